// allpairs.cuh — Allpairs skeleton:
//   allpairs(+)(A, B) = C,  C[i][j] = A_i (+) B_j   (rows of the n x d matrix A
//   and the m x d matrix B)
//
// Two forms:
//  * generic (SKL_AP_ZR 0): the customising function gets two row pointers and
//    d, `TOUT f(const TIN* a, const TIN* b, int d)` (reading A35).  A block
//    computes a 16 x 16 tile of C, one element per thread, with the 16 A rows
//    and 16 B rows it needs staged in shared memory (row pitch d+1: no bank
//    conflicts) when they fit, else read from global memory;
//  * zip-reduce (SKL_AP_ZR 1): C[i][j] = fold((+), zip((x), A_i, B_j)), the
//    left fold acc = z_0, acc = acc (+) z_k (no identity, A10) of two customising
//    functions (reading A36: the SkelCL line of work specialises Allpairs this
//    way).  Register-tiled like an SGEMM on the FP32 pipes: a 64 x 64 tile of C
//    per block, 4 x 4 per thread, k-slices of 16 staged k-major in shared memory.
//    Every C element is folded in k order, so results equal the oracle's
//    sequential fold bit for bit (-fmad=false).  No tensor cores: the operators
//    are arbitrary (the dotProduct / matrix-multiply special case of Eq. (2)
//    would belong on tcgen05; out of scope here).
// Configuration: SKL_TIN, SKL_TOUT, SKL_BLOCK (256), SKL_AP_ZR, SKL_FUNC or
// SKL_ZFUNC / SKL_RFUNC.

#if SKL_AP_ZR
#define AP_BM 64
#define AP_BN 64
#define AP_BK 16
extern "C" __global__ void __launch_bounds__(256)
skl_ap_zr(const SKL_TIN* __restrict__ A, const SKL_TIN* __restrict__ B, SKL_TOUT* __restrict__ Cm,
          long n, long m, long d) {
  __shared__ SKL_TIN As[AP_BK][AP_BM + 1];  // +1: the transposing stores hit distinct banks
  __shared__ SKL_TIN Bs[AP_BK][AP_BN + 1];
  const int tx = threadIdx.x & 15, ty = threadIdx.x >> 4;
  const long i0 = (long)blockIdx.y * AP_BM, j0 = (long)blockIdx.x * AP_BN;
  SKL_TOUT acc[4][4];
  for (long k0 = 0; k0 < d; k0 += AP_BK) {
    // stage A[i0 .. i0+63][k0 .. k0+15] and B likewise, k-major (4 elements each)
#pragma unroll
    for (int q = 0; q < 4; ++q) {
      const int e = threadIdx.x + q * 256;  // 0 .. 1023
      const int r = e >> 4, c = e & 15;     // row within the tile, k within the slice
      const long k = k0 + c;
      SKL_TIN va, vb;
      if (i0 + r < n && k < d) va = A[(i0 + r) * d + k];
      if (j0 + r < m && k < d) vb = B[(j0 + r) * d + k];
      As[c][r] = va;
      Bs[c][r] = vb;
    }
    __syncthreads();
    const int kn = d - k0 < AP_BK ? (int)(d - k0) : AP_BK;
#pragma unroll
    for (int kk = 0; kk < AP_BK; ++kk) {
      if (kk < kn) {
        SKL_TIN a[4], b[4];
#pragma unroll
        for (int r = 0; r < 4; ++r) a[r] = As[kk][ty * 4 + r];
#pragma unroll
        for (int c = 0; c < 4; ++c) b[c] = Bs[kk][tx * 4 + c];
        const bool first = (k0 == 0 && kk == 0);
#pragma unroll
        for (int r = 0; r < 4; ++r)
#pragma unroll
          for (int c = 0; c < 4; ++c) {
            const SKL_TOUT z = SKL_ZFUNC(a[r], b[c]);
            acc[r][c] = first ? z : SKL_RFUNC(acc[r][c], z);
          }
      }
    }
    __syncthreads();
  }
#pragma unroll
  for (int r = 0; r < 4; ++r) {
    const long i = i0 + ty * 4 + r;
    if (i >= n) continue;
#pragma unroll
    for (int c = 0; c < 4; ++c) {
      const long j = j0 + tx * 4 + c;
      if (j < m) Cm[i * m + j] = acc[r][c];
    }
  }
}
#else
extern "C" __global__ void __launch_bounds__(256)
skl_ap_gen(const SKL_TIN* __restrict__ A, const SKL_TIN* __restrict__ B, SKL_TOUT* __restrict__ Cm,
           long n, long m, long d, int use_smem) {
  extern __shared__ __align__(16) unsigned char skl_ap_raw[];
  SKL_TIN* sA = (SKL_TIN*)skl_ap_raw;            // [16][d+1]
  SKL_TIN* sB = sA + 16 * (d + 1);               // [16][d+1]
  const int tx = threadIdx.x & 15, ty = threadIdx.x >> 4;
  const long i0 = (long)blockIdx.y * 16, j0 = (long)blockIdx.x * 16;
  if (use_smem) {
    for (long e = threadIdx.x; e < 16 * d; e += 256) {
      const long r = e / d, k = e - r * d;
      if (i0 + r < n) sA[r * (d + 1) + k] = A[(i0 + r) * d + k];
      if (j0 + r < m) sB[r * (d + 1) + k] = B[(j0 + r) * d + k];
    }
    __syncthreads();
  }
  const long i = i0 + ty, j = j0 + tx;
  if (i < n && j < m) {
    const SKL_TIN* a = use_smem ? sA + ty * (d + 1) : A + i * d;
    const SKL_TIN* b = use_smem ? sB + tx * (d + 1) : B + j * d;
    Cm[i * m + j] = SKL_FUNC((SKL_TIN*)a, (SKL_TIN*)b, (int)d);
  }
}
#endif
