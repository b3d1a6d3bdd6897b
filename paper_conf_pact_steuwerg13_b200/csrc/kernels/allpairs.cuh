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

#if SKL_AP_FAST
// 4-byte inputs, d % 4 == 0, 16-byte aligned rows: a 128 x 128 tile of C per
// block, 8 x 8 per thread (rows ty + 16 r, columns tx + 16 c: consecutive
// lanes read consecutive rows, so the 16-byte shared loads are conflict-free
// with an 80-byte row pitch), k-slices of 16 staged row-major by cp.async into
// a double buffer; per k-quad a thread issues 16 LDS.128 for 512 FP32 ops.
// Every accumulator is still folded in k order (bit-exact with the oracle).
#define AQ_BM 128
#ifdef SKL_AP_BK
#define AQ_BK SKL_AP_BK
#else
#define AQ_BK 16
#endif
#define AQ_P (AQ_BK + 4)
#define AQ_CPR (AQ_BK / 4)   // 16-byte chunks per staged row
union SklAp4 {
  uint4 q;
  SKL_TIN e[4];
};
__device__ __forceinline__ void skl_ap_cp16(void* smem, const void* g) {
  const unsigned sa = (unsigned)__cvta_generic_to_shared(smem);
  asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" ::"r"(sa), "l"(g) : "memory");
}
// 16 k of a staged slice, from column koff (unrolled body; deeper slices loop over it)
template <bool FIRST, int TC>
__device__ __forceinline__ void skl_ap_slice16(SKL_TOUT (&acc)[8][TC], const SKL_TIN* As, const SKL_TIN* Bs,
                                               int tx, int ty, int koff) {
#pragma unroll
  for (int kq = 0; kq < 16; kq += 4) {
    SklAp4 a[8];
#pragma unroll
    for (int r = 0; r < 8; ++r) a[r].q = *(const uint4*)&As[(ty + 16 * r) * AQ_P + koff + kq];
#pragma unroll
    for (int c = 0; c < TC; ++c) {
      SklAp4 b;
      b.q = *(const uint4*)&Bs[(tx + 16 * c) * AQ_P + koff + kq];
#pragma unroll
      for (int j = 0; j < 4; ++j)
#pragma unroll
        for (int r = 0; r < 8; ++r) {
          const SKL_TOUT z = SKL_ZFUNC(a[r].e[j], b.e[j]);
          acc[r][c] = (FIRST && kq == 0 && j == 0) ? z : SKL_RFUNC(acc[r][c], z);
        }
    }
  }
}
template <bool FIRST, int TC>
__device__ __forceinline__ void skl_ap_slice(SKL_TOUT (&acc)[8][TC], const SKL_TIN* As, const SKL_TIN* Bs,
                                             int tx, int ty) {
  skl_ap_slice16<FIRST, TC>(acc, As, Bs, tx, ty, 0);
#pragma unroll 1
  for (int k16 = 16; k16 < AQ_BK; k16 += 16) skl_ap_slice16<false, TC>(acc, As, Bs, tx, ty, k16);
}
// One 128 x (16 TC) tile of C at (i0, j0) per block of 256 threads, 8 x TC per
// thread; sm holds 2 * (128 + 16 TC) * AQ_P elements.
#define AQ_STAGE(TC) ((AQ_BM + 16 * (TC)) * AQ_P)
template <int TC>
__device__ __forceinline__ void skl_ap_tile(const SKL_TIN* __restrict__ A, const SKL_TIN* __restrict__ B,
                                            SKL_TOUT* __restrict__ Cm, long n, long m, long d, long i0, long j0,
                                            SKL_TIN* sm) {
  constexpr int BN = 16 * TC;                      // tile columns (rows of B)
  constexpr int STAGE = AQ_STAGE(TC);
  const int tx = threadIdx.x & 15, ty = threadIdx.x >> 4;
  const long nfull = d / AQ_BK;
  // chunk q of a (rows x 16) slab: row q / 4, k-quad q % 4 (rows beyond n / m
  // are clamped to the last one: loaded, never stored)
  constexpr int HA = AQ_BM * AQ_CPR / 256, HB = BN * AQ_CPR / 256;   // chunks per thread
  long ra[HA], rb[HB];
#pragma unroll
  for (int h = 0; h < HA; ++h) {
    const int r = (threadIdx.x + h * 256) / AQ_CPR;
    ra[h] = (i0 + r < n ? i0 + r : n - 1) * d;
  }
#pragma unroll
  for (int h = 0; h < HB; ++h) {
    const int r = (threadIdx.x + h * 256) / AQ_CPR;
    rb[h] = (j0 + r < m ? j0 + r : m - 1) * d;
  }
  auto stage = [&](int st, long k0) {
    SKL_TIN* As = sm + st * STAGE;
    SKL_TIN* Bs = As + AQ_BM * AQ_P;
#pragma unroll
    for (int h = 0; h < HA; ++h) {
      const int q = threadIdx.x + h * 256, r = q / AQ_CPR, kq = (q % AQ_CPR) * 4;
      skl_ap_cp16(&As[r * AQ_P + kq], A + ra[h] + k0 + kq);
    }
#pragma unroll
    for (int h = 0; h < HB; ++h) {
      const int q = threadIdx.x + h * 256, r = q / AQ_CPR, kq = (q % AQ_CPR) * 4;
      skl_ap_cp16(&Bs[r * AQ_P + kq], B + rb[h] + k0 + kq);
    }
  };
  SKL_TOUT acc[8][TC];
  if (nfull > 0) stage(0, 0);
  asm volatile("cp.async.commit_group;" ::: "memory");
  for (long s = 0; s < nfull; ++s) {
    if (s + 1 < nfull) stage((int)((s + 1) & 1), (s + 1) * AQ_BK);
    asm volatile("cp.async.commit_group;" ::: "memory");
    asm volatile("cp.async.wait_group 1;" ::: "memory");
    __syncthreads();
    const SKL_TIN* As = sm + (s & 1) * STAGE;
    if (s == 0) skl_ap_slice<true, TC>(acc, As, As + AQ_BM * AQ_P, tx, ty);
    else skl_ap_slice<false, TC>(acc, As, As + AQ_BM * AQ_P, tx, ty);
    __syncthreads();  // the next stage() overwrites this buffer
  }
  // tail k-slice (d % 16 elements): scalar, guarded
  const int kt = (int)(d - nfull * AQ_BK);
  if (kt > 0) {
    asm volatile("cp.async.wait_group 0;" ::: "memory");
    SKL_TIN* As = sm;
    SKL_TIN* Bs = As + AQ_BM * AQ_P;
    const long k0 = nfull * AQ_BK;
    for (int e = threadIdx.x; e < (AQ_BM + BN) * AQ_BK; e += 256) {
      const int r = e / AQ_BK, k = e % AQ_BK;
      if (k >= kt) continue;
      if (r < AQ_BM) {
        const long ia = i0 + r < n ? i0 + r : n - 1;
        As[r * AQ_P + k] = A[ia * d + k0 + k];
      } else {
        const long jb = j0 + (r - AQ_BM) < m ? j0 + (r - AQ_BM) : m - 1;
        Bs[(r - AQ_BM) * AQ_P + k] = B[jb * d + k0 + k];
      }
    }
    __syncthreads();
    for (int k = 0; k < kt; ++k)
#pragma unroll
      for (int r = 0; r < 8; ++r)
#pragma unroll
        for (int c = 0; c < TC; ++c) {
          const SKL_TOUT z = SKL_ZFUNC(As[(ty + 16 * r) * AQ_P + k], Bs[(tx + 16 * c) * AQ_P + k]);
          acc[r][c] = (nfull == 0 && k == 0) ? z : SKL_RFUNC(acc[r][c], z);
        }
  }
#pragma unroll
  for (int r = 0; r < 8; ++r) {
    const long i = i0 + ty + 16 * r;
    if (i >= n) continue;
#pragma unroll
    for (int c = 0; c < TC; ++c) {
      const long j = j0 + tx + 16 * c;
      if (j < m) Cm[i * m + j] = acc[r][c];
    }
  }
}
// 128 x 128 tiles (2 blocks per SM) and 128 x 64 tiles (3 blocks per SM, twice
// the tiles: the host picks the one whose tile count fills the waves better)
extern "C" __global__ void __launch_bounds__(256, 2)
skl_ap_zr8(const SKL_TIN* __restrict__ A, const SKL_TIN* __restrict__ B, SKL_TOUT* __restrict__ Cm,
           long n, long m, long d) {
  extern __shared__ __align__(16) unsigned char skl_ap_dyn[];   // 2 * AQ_STAGE(8) elements
  skl_ap_tile<8>(A, B, Cm, n, m, d, (long)blockIdx.y * AQ_BM, (long)blockIdx.x * 128, (SKL_TIN*)skl_ap_dyn);
}
extern "C" __global__ void __launch_bounds__(256, 3)
skl_ap_zr4(const SKL_TIN* __restrict__ A, const SKL_TIN* __restrict__ B, SKL_TOUT* __restrict__ Cm,
           long n, long m, long d) {
  extern __shared__ __align__(16) unsigned char skl_ap_dyn[];   // 2 * AQ_STAGE(4) elements
  skl_ap_tile<4>(A, B, Cm, n, m, d, (long)blockIdx.y * AQ_BM, (long)blockIdx.x * 64, (SKL_TIN*)skl_ap_dyn);
}
// Wave-quantisation fix: the 128 x 128 tiles (row-major, tiles_x per row) that
// fill whole waves run as such (blocks 0 .. nwide-1); each tile of the last,
// partial wave is split into two 128 x 64 halves (blocks nwide ..), so the
// last wave has twice the blocks, each half the work.  Every C element is still
// folded in k order by one thread (bit-exact).
extern "C" __global__ void __launch_bounds__(256, 2)
skl_ap_zrh(const SKL_TIN* __restrict__ A, const SKL_TIN* __restrict__ B, SKL_TOUT* __restrict__ Cm,
           long n, long m, long d, long nwide, long tiles_x) {
  extern __shared__ __align__(16) unsigned char skl_ap_dyn[];   // 2 * AQ_STAGE(8) elements
  SKL_TIN* sm = (SKL_TIN*)skl_ap_dyn;
  const long b = blockIdx.x;
  if (b < nwide) {
    skl_ap_tile<8>(A, B, Cm, n, m, d, (b / tiles_x) * AQ_BM, (b % tiles_x) * 128, sm);
  } else {
    const long t = nwide + (b - nwide) / 2;
    const long j0 = (t % tiles_x) * 128 + ((b - nwide) & 1) * 64;
    if (j0 < m) skl_ap_tile<4>(A, B, Cm, n, m, d, (t / tiles_x) * AQ_BM, j0, sm);
  }
}
#endif
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
