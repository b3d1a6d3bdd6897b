// reduce.cuh — Reduce skeleton:  red (+) [v1..vn] = v1 (+) ... (+) vn
//
// (+) is only associative: no identity element exists and operands are
// never reordered (reading A10).  Order-preserving design for sm_100a:
//  * every warp owns one contiguous segment of the vector, blocks own
//    consecutive runs of warps, so a left-to-right fold of warp results, then of
//    block results, is the vector's fold;
//  * a warp streams tiles of 32 lanes x SKL_RVEC elements (one 16-byte load per
//    lane, SKL_RU tiles in flight); each lane folds its SKL_RVEC consecutive
//    elements left to right, then an order-preserving shuffle tree folds the 32
//    lane values (skl_warp_fold; partial tiles skip the missing lanes);
//  * block partials are folded in order by the last block to finish (one launch,
//    no second kernel): ticket counter + __threadfence.
// Configuration: SKL_T, SKL_FUNC, SKL_BLOCK, SKL_RVEC, SKL_RU.
#define SKL_NW (SKL_BLOCK / 32)
#define SKL_RTILE (32 * SKL_RVEC)

template <int RVEC>
__device__ __forceinline__ void skl_reduce_body(const SKL_T* __restrict__ in, skl_u64 n, skl_u64 wseg,
                                                SKL_T* partials, unsigned* counter, SKL_T* result) {
  SklOp op;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const skl_u64 w = (skl_u64)blockIdx.x * SKL_NW + warp;
  const skl_u64 lo = w * wseg;
  const skl_u64 hi = lo + wseg < n ? lo + wseg : n;
  bool has = false;
  SKL_T acc;
  for (skl_u64 t = lo; t < hi; t += (skl_u64)SKL_RTILE * SKL_RU) {
    SKL_T x[SKL_RU][RVEC];
    int cnt[SKL_RU];
#pragma unroll
    for (int u = 0; u < SKL_RU; ++u) {
      const skl_u64 e = t + (skl_u64)u * SKL_RTILE + (skl_u64)lane * RVEC;
      cnt[u] = e >= hi ? 0 : (hi - e >= (skl_u64)RVEC ? RVEC : (int)(hi - e));
      if (RVEC > 1 && cnt[u] == RVEC) {
        SklChunk<SKL_T, RVEC> ch;
        ch.q[0] = skl_ld16(in + e);
#pragma unroll
        for (int k = 0; k < RVEC; ++k) x[u][k] = ch.e[k];
      } else {
#pragma unroll
        for (int k = 0; k < RVEC; ++k)
          if (k < cnt[u]) x[u][k] = in[e + k];
      }
    }
#pragma unroll
    for (int u = 0; u < SKL_RU; ++u) {
      const skl_u64 tl = t + (skl_u64)u * SKL_RTILE;
      if (tl >= hi) break;
      SKL_T v = x[u][0];
#pragma unroll
      for (int k = 1; k < RVEC; ++k)
        if (k < cnt[u]) v = op(v, x[u][k]);
      const skl_u64 rem = hi - tl;
      const int nv = rem >= (skl_u64)SKL_RTILE ? 32 : (int)((rem + RVEC - 1) / RVEC);
      v = skl_warp_fold(v, nv, op);
      v = skl_shfl(v, 0);
      acc = has ? op(acc, v) : v;
      has = true;
    }
  }
  // block: fold warp results in warp order (empty warps are a suffix)
  __shared__ SKL_T s_w[SKL_NW];
  __shared__ int s_h[SKL_NW];
  __shared__ int s_last;
  if (lane == 0) {
    s_h[warp] = has;
    if (has) s_w[warp] = acc;
  }
  __syncthreads();
  if (threadIdx.x == 0) {
    SKL_T b = s_w[0];
    for (int i = 1; i < SKL_NW; ++i)
      if (s_h[i]) b = op(b, s_w[i]);
    if (gridDim.x == 1) {
      *result = b;
    } else {
      partials[blockIdx.x] = b;
      __threadfence();
      const unsigned ticket = atomicAdd(counter, 1u);
      s_last = (ticket == gridDim.x - 1);
    }
  }
  if (gridDim.x == 1) return;
  __syncthreads();
  if (!s_last || warp != 0) return;
  // last block: fold the block partials in block order
  __threadfence();
  bool h2 = false;
  SKL_T a2;
  for (unsigned b0 = 0; b0 < gridDim.x; b0 += 32) {
    const unsigned nb = gridDim.x - b0 < 32 ? gridDim.x - b0 : 32;
    SKL_T v;
    if ((unsigned)lane < nb) v = skl_ldcg(partials + b0 + lane);
    v = skl_warp_fold(v, (int)nb, op);
    v = skl_shfl(v, 0);
    a2 = h2 ? op(a2, v) : v;
    h2 = true;
  }
  if (lane == 0) {
    *result = a2;
    *counter = 0u;  // ready for the next launch (stream-ordered)
  }
}

extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_reduce_vec(const SKL_T* __restrict__ in, skl_u64 n, skl_u64 wseg, SKL_T* partials,
               unsigned* counter, SKL_T* result) {
  skl_reduce_body<SKL_RVEC>(in, n, wseg, partials, counter, result);
}
extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_reduce_sc(const SKL_T* __restrict__ in, skl_u64 n, skl_u64 wseg, SKL_T* partials,
              unsigned* counter, SKL_T* result) {
  skl_reduce_body<1>(in, n, wseg, partials, counter, result);
}

// Ordered fold of `nrep` staged values per element (copy(+) -> block combine,
// reading A25; and the cross-GPU fold of Reduce partials): out[i] =
// s[0][i] (+) s[1][i] (+) ... (+) s[nrep-1][i], GPU order.
extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_combine(const SKL_T* __restrict__ staging, skl_u64 stride, int nrep, SKL_T* __restrict__ out,
            skl_u64 n) {
  SklOp op;
  for (skl_u64 i = (skl_u64)blockIdx.x * SKL_BLOCK + threadIdx.x; i < n;
       i += (skl_u64)gridDim.x * SKL_BLOCK) {
    SKL_T a = staging[i];
    for (int r = 1; r < nrep; ++r) a = op(a, staging[(skl_u64)r * stride + i]);
    out[i] = a;
  }
}
