// scan.cuh — Scan skeleton, inclusive (reading A9):
//   scan (+) [v1..vn] = [v1, v1 (+) v2, ..., v1 (+) ... (+) vn]
//
// Single-pass decoupled look-back (Merrill & Garland) for an operator that is
// only associative: no identity is ever used, and every
// combination keeps the left operand at the lower index (A10).
//  * one block per tile of SKL_BLOCK x SKL_ITEMS elements; tile t = blockIdx.x
//    (blocks are dispatched in index order, so a tile only waits on tiles that
//    are already resident or done);
//  * vector path: the tile moves global<->smem as coalesced 16-byte chunks with
//    an XOR swizzle pos(c) = c ^ ((c >> 3) & 7) that keeps both the striped
//    global-order accesses and the per-thread blocked accesses (SKL_CH
//    consecutive chunks per thread) free of shared-memory bank conflicts;
//  * per thread: sequential inclusive scan of SKL_ITEMS registers; per warp:
//    shuffle scan of thread totals; per block: fold of warp totals;
//  * tile status = (epoch << 2 | {1: aggregate, 2: inclusive prefix}) with
//    release/acquire ordering; warp 0 looks back 32 predecessors at a time and
//    folds them right-to-left-in-lanes (= left-to-right in the vector);
//  * multi-GPU carry-in: tile 0 of GPU g starts from
//    carry[0] (+) ... (+) carry[ncarry-1], the totals of GPUs 0..g-1.
// Configuration: SKL_T, SKL_FUNC, SKL_BLOCK, SKL_ITEMS, SKL_CH (16-byte chunks
// per thread on the vector path; 0 = generic path only).
#define SKL_NW (SKL_BLOCK / 32)
#define SKL_TILE (SKL_BLOCK * SKL_ITEMS)

__device__ __forceinline__ unsigned skl_swz(unsigned c) { return c ^ ((c >> 3) & 7u); }

// Tile-level exclusive prefix via decoupled look-back (called by warp 0).
// Publishes this tile's aggregate first and its inclusive prefix last.
__device__ __forceinline__ void skl_lookback(unsigned tile, const SKL_T& agg, unsigned* flags,
                                             SKL_T* aggs, SKL_T* incls, unsigned epoch,
                                             const SKL_T* carry, int ncarry, SKL_T* s_excl,
                                             int* s_has) {
  SklOp op;
  const int lane = threadIdx.x & 31;
  if (tile == 0) {
    if (lane == 0) {
      if (ncarry > 0) {
        SKL_T c = carry[0];
        for (int i = 1; i < ncarry; ++i) c = op(c, carry[i]);
        incls[0] = op(c, agg);
        *s_excl = c;
        *s_has = 1;
      } else {
        incls[0] = agg;
        *s_has = 0;
      }
      skl_st_release(&flags[0], (epoch << 2) | 2u);
    }
    return;
  }
  if (lane == 0) {
    aggs[tile] = agg;
    skl_st_release(&flags[tile], (epoch << 2) | 1u);
  }
  bool have = false;
  SKL_T acc;
  long base = (long)tile - 1;
  while (true) {
    const long j = base - lane;
    unsigned st;
    do {
      const unsigned f = j >= 0 ? skl_ld_acquire(&flags[j]) : 0u;
      st = (f >> 2) == epoch ? (f & 3u) : 0u;
    } while (__any_sync(SKL_FULL, j >= 0 && st == 0u));
    const unsigned pm = __ballot_sync(SKL_FULL, j >= 0 && st == 2u);
    const int p = pm ? __ffs(pm) - 1 : 31;
    SKL_T v;
    if (lane <= p && j >= 0) v = (pm && lane == p) ? skl_ldcg(incls + j) : skl_ldcg(aggs + j);
    // lanes p..0 are tiles j = base-p .. base: fold with the higher lane on the left
#pragma unroll
    for (int s = 1; s < 32; s <<= 1) {
      SKL_T o = skl_shfl_down(v, s);
      if (lane + s <= p) v = op(o, v);
    }
    v = skl_shfl(v, 0);
    acc = have ? op(v, acc) : v;
    have = true;
    if (pm) break;
    base -= 32;
  }
  if (lane == 0) {
    incls[tile] = op(acc, agg);
    skl_st_release(&flags[tile], (epoch << 2) | 2u);
    *s_excl = acc;
    *s_has = 1;
  }
}

// Shared body: items[] holds this thread's (blocked) elements, cnt of them valid.
// On return items[k] holds the inclusive scan value of element t*ITEMS+k.
__device__ __forceinline__ void skl_scan_tile(SKL_T (&items)[SKL_ITEMS], int cnt, int nthr_valid,
                                              unsigned* flags, SKL_T* aggs, SKL_T* incls,
                                              unsigned epoch, const SKL_T* carry, int ncarry) {
  SklOp op;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  // 1. sequential inclusive scan inside the thread
  SKL_T v = items[0];
#pragma unroll
  for (int k = 1; k < SKL_ITEMS; ++k)
    if (k < cnt) {
      items[k] = op(items[k - 1], items[k]);
      v = items[k];
    }
  // 2. warp inclusive scan of thread totals (valid threads are a prefix)
#pragma unroll
  for (int s = 1; s < 32; s <<= 1) {
    SKL_T o = skl_shfl_up(v, s);
    if (lane >= s) v = op(o, v);
  }
  SKL_T lane_excl = skl_shfl_up(v, 1);
  __shared__ SKL_T s_wt[SKL_NW];
  __shared__ SKL_T s_wex[SKL_NW];
  __shared__ SKL_T s_agg, s_excl;
  __shared__ int s_has;
  const int wvalid = nthr_valid - warp * 32;  // valid threads in this warp
  if (wvalid > 0 && lane == (wvalid >= 32 ? 31 : wvalid - 1)) s_wt[warp] = v;
  __syncthreads();
  // 3. block: exclusive prefixes of warp totals, tile aggregate
  if (threadIdx.x == 0) {
    const int nwv = (nthr_valid + 31) / 32;
    SKL_T a = s_wt[0];
    for (int w = 1; w < nwv; ++w) {
      s_wex[w] = a;
      a = op(a, s_wt[w]);
    }
    s_agg = a;
  }
  __syncthreads();
  // 4. look-back for the tile prefix
  if (warp == 0) {
    SKL_T agg = s_agg;
    skl_lookback(blockIdx.x, agg, flags, aggs, incls, epoch, carry, ncarry, &s_excl, &s_has);
  }
  __syncthreads();
  // 5. this thread's exclusive prefix = tile prefix (+) warp prefix (+) lane prefix
  bool hp = s_has != 0;
  SKL_T pre;
  if (hp) pre = s_excl;
  if (warp > 0) {
    pre = hp ? op(pre, s_wex[warp]) : s_wex[warp];
    hp = true;
  }
  if (lane > 0) {
    pre = hp ? op(pre, lane_excl) : lane_excl;
    hp = true;
  }
  if (hp) {
#pragma unroll
    for (int k = 0; k < SKL_ITEMS; ++k)
      if (k < cnt) items[k] = op(pre, items[k]);
  }
}

#if SKL_CH > 0
// Vector path: sizeof(T) divides 16, in/out 16-byte aligned.
#define SKL_EPC (16 / (int)sizeof(SKL_T))  // elements per chunk
extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_scan_vec(const SKL_T* __restrict__ in, SKL_T* __restrict__ out, skl_u64 n, unsigned* flags,
             SKL_T* aggs, SKL_T* incls, unsigned epoch, const SKL_T* carry, int ncarry) {
  __shared__ uint4 sm[SKL_BLOCK * SKL_CH];
  const skl_u64 tlo = (skl_u64)blockIdx.x * SKL_TILE;
  const int nvalid = n - tlo >= (skl_u64)SKL_TILE ? SKL_TILE : (int)(n - tlo);
  const char* gin = (const char*)(in + tlo);
  if (nvalid == SKL_TILE) {
#pragma unroll
    for (int i = 0; i < SKL_CH; ++i) {
      const unsigned c = i * SKL_BLOCK + threadIdx.x;
      sm[skl_swz(c)] = skl_ld16(gin + 16 * (skl_u64)c);
    }
  } else {
    for (int e = threadIdx.x; e < nvalid; e += SKL_BLOCK) {
      SKL_T* slot = (SKL_T*)&sm[skl_swz(e / SKL_EPC)] + (e % SKL_EPC);
      *slot = in[tlo + e];
    }
  }
  __syncthreads();
  SklChunk<SKL_T, SKL_ITEMS> my;
#pragma unroll
  for (int k = 0; k < SKL_CH; ++k) my.q[k] = sm[skl_swz(threadIdx.x * SKL_CH + k)];
  SKL_T items[SKL_ITEMS];
#pragma unroll
  for (int k = 0; k < SKL_ITEMS; ++k) items[k] = my.e[k];
  const int first = threadIdx.x * SKL_ITEMS;
  const int cnt = nvalid - first >= SKL_ITEMS ? SKL_ITEMS : (nvalid - first > 0 ? nvalid - first : 0);
  const int nthr = (nvalid + SKL_ITEMS - 1) / SKL_ITEMS;
  skl_scan_tile(items, cnt, nthr, flags, aggs, incls, epoch, carry, ncarry);
#pragma unroll
  for (int k = 0; k < SKL_ITEMS; ++k) my.e[k] = items[k];
  __syncthreads();  // everyone has read sm
#pragma unroll
  for (int k = 0; k < SKL_CH; ++k) sm[skl_swz(threadIdx.x * SKL_CH + k)] = my.q[k];
  __syncthreads();
  char* gout = (char*)(out + tlo);
  if (nvalid == SKL_TILE) {
#pragma unroll
    for (int i = 0; i < SKL_CH; ++i) {
      const unsigned c = i * SKL_BLOCK + threadIdx.x;
      skl_st16(gout + 16 * (skl_u64)c, sm[skl_swz(c)]);
    }
  } else {
    for (int e = threadIdx.x; e < nvalid; e += SKL_BLOCK)
      out[tlo + e] = *((const SKL_T*)&sm[skl_swz(e / SKL_EPC)] + (e % SKL_EPC));
  }
}
#endif

// Generic path: any element size / alignment (blocked layout through smem).
extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_scan_sc(const SKL_T* __restrict__ in, SKL_T* __restrict__ out, skl_u64 n, unsigned* flags,
            SKL_T* aggs, SKL_T* incls, unsigned epoch, const SKL_T* carry, int ncarry) {
  __shared__ __align__(16) unsigned char sm_raw[SKL_TILE * sizeof(SKL_T)];
  SKL_T* sm_u = (SKL_T*)sm_raw;
  const skl_u64 tlo = (skl_u64)blockIdx.x * SKL_TILE;
  const int nvalid = n - tlo >= (skl_u64)SKL_TILE ? SKL_TILE : (int)(n - tlo);
  for (int e = threadIdx.x; e < nvalid; e += SKL_BLOCK) sm_u[e] = in[tlo + e];
  __syncthreads();
  SKL_T items[SKL_ITEMS];
  const int first = threadIdx.x * SKL_ITEMS;
#pragma unroll
  for (int k = 0; k < SKL_ITEMS; ++k)
    if (first + k < nvalid) items[k] = sm_u[first + k];
  const int cnt = nvalid - first >= SKL_ITEMS ? SKL_ITEMS : (nvalid - first > 0 ? nvalid - first : 0);
  const int nthr = (nvalid + SKL_ITEMS - 1) / SKL_ITEMS;
  skl_scan_tile(items, cnt, nthr, flags, aggs, incls, epoch, carry, ncarry);
  __syncthreads();
#pragma unroll
  for (int k = 0; k < SKL_ITEMS; ++k)
    if (k < cnt) sm_u[first + k] = items[k];
  __syncthreads();
  for (int e = threadIdx.x; e < nvalid; e += SKL_BLOCK) out[tlo + e] = sm_u[e];
}
