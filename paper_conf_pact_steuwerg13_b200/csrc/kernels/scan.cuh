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

// ---- tile status words (decoupled look-back) ---------------------------------
// SKL_PACKED (sizeof(T) <= 4, like CUB): one 64-bit word per tile holds
// (value bits << 32 | epoch << 2 | state); a relaxed 64-bit load sees the value
// together with its flag, so neither side needs a fence.  (ld.acquire.gpu makes
// ptxas emit CCTL.IVALL - an L1 invalidate - on every spin iteration; measured as
// the top stall of the first version.)  Otherwise: separate value arrays, a
// relaxed flag spin, and one fence per look-back round before the value loads.
// States: 0 = not yet published (or an older epoch), 1 = aggregate, 2 = prefix.
__device__ __forceinline__ unsigned long long skl_ld_relaxed64(const unsigned long long* p) {
  unsigned long long v;
  asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void skl_st_relaxed64(unsigned long long* p, unsigned long long v) {
  asm volatile("st.relaxed.gpu.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ unsigned skl_ld_relaxed32(const unsigned* p) {
  unsigned v;
  asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}

// Status words are SKL_FSTRIDE x 8 bytes apart (default 128 B: one L2 line per
// tile) so that the blocks polling the look-back frontier spread over L2 slices
// instead of hammering the one line that holds 16 neighbouring tiles' words.
#ifndef SKL_FSTRIDE
#define SKL_FSTRIDE 16
#endif
#ifndef SKL_SPIN_NS
#define SKL_SPIN_NS 0
#endif

#ifndef SKL_LBW
#define SKL_LBW 3
#endif

#if SKL_PACKED
// one look at tile j's status: 0 if not published yet, else state (*v = value)
__device__ __forceinline__ unsigned skl_status_try(const unsigned* flags, const SKL_T* aggs,
                                                   const SKL_T* incls, long j, unsigned epoch, SKL_T* v) {
  const unsigned long long w = skl_ld_relaxed64((const unsigned long long*)flags + (skl_u64)j * SKL_FSTRIDE);
  const unsigned st = ((unsigned)w >> 2) == epoch ? ((unsigned)w & 3u) : 0u;
  if (st) {
    const unsigned bits = (unsigned)(w >> 32);
    memcpy(v, &bits, sizeof(SKL_T));
  }
  (void)aggs;
  (void)incls;
  return st;
}
__device__ __forceinline__ void skl_publish(unsigned* flags, SKL_T* aggs, SKL_T* incls, unsigned tile,
                                            unsigned epoch, unsigned state, const SKL_T& v) {
  unsigned bits = 0;
  memcpy(&bits, &v, sizeof(SKL_T));
  skl_st_relaxed64((unsigned long long*)flags + (skl_u64)tile * SKL_FSTRIDE,
                   ((unsigned long long)bits << 32) | (unsigned long long)((epoch << 2) | state));
  (void)aggs;
  (void)incls;
}
// spin until tile j is published; returns its state, *v its value
__device__ __forceinline__ unsigned skl_status(const unsigned* flags, const SKL_T* aggs,
                                               const SKL_T* incls, long j, unsigned epoch, SKL_T* v) {
  unsigned long long w;
  unsigned st;
  do {
    w = skl_ld_relaxed64((const unsigned long long*)flags + (skl_u64)j * SKL_FSTRIDE);
    st = ((unsigned)w >> 2) == epoch ? ((unsigned)w & 3u) : 0u;
    if (st == 0u) __nanosleep(SKL_SPIN_NS);
  } while (st == 0u);
  const unsigned bits = (unsigned)(w >> 32);
  memcpy(v, &bits, sizeof(SKL_T));
  (void)aggs;
  (void)incls;
  return st;
}
#else
__device__ __forceinline__ unsigned skl_status_try(const unsigned* flags, const SKL_T* aggs,
                                                   const SKL_T* incls, long j, unsigned epoch, SKL_T* v) {
  const unsigned f = skl_ld_relaxed32(&flags[(skl_u64)j * 2 * SKL_FSTRIDE]);
  const unsigned st = (f >> 2) == epoch ? (f & 3u) : 0u;
  if (st) {
    __threadfence();  // acquire
    *v = st == 2u ? skl_ldcg(incls + j) : skl_ldcg(aggs + j);
  }
  return st;
}
__device__ __forceinline__ void skl_publish(unsigned* flags, SKL_T* aggs, SKL_T* incls, unsigned tile,
                                            unsigned epoch, unsigned state, const SKL_T& v) {
  if (state == 1u) aggs[tile] = v;
  else incls[tile] = v;
  skl_st_release(&flags[(skl_u64)tile * 2 * SKL_FSTRIDE], (epoch << 2) | state);
}
__device__ __forceinline__ unsigned skl_status(const unsigned* flags, const SKL_T* aggs,
                                               const SKL_T* incls, long j, unsigned epoch, SKL_T* v) {
  unsigned f, st;
  do {
    f = skl_ld_relaxed32(&flags[(skl_u64)j * 2 * SKL_FSTRIDE]);
    st = (f >> 2) == epoch ? (f & 3u) : 0u;
    if (st == 0u) __nanosleep(SKL_SPIN_NS);
  } while (st == 0u);
  __threadfence();  // acquire: the value written before the release is visible now
  *v = st == 2u ? skl_ldcg(incls + j) : skl_ldcg(aggs + j);
  return st;
}
#endif

// Block-wide look-back: every thread watches one predecessor tile, so one L2
// round trip covers SKL_BLOCK tiles (a warp-wide window advances the inclusive-
// prefix frontier only 32 tiles per round trip).  Called by all threads; *s_agg
// is this tile's aggregate.  Results: *s_excl / *s_has (tile's exclusive prefix).
__device__ __forceinline__ void skl_lookback_block(unsigned tile, unsigned* flags, SKL_T* aggs,
                                                   SKL_T* incls, unsigned epoch, const SKL_T* carry,
                                                   int ncarry, const SKL_T* s_agg, SKL_T* s_excl,
                                                   int* s_has, bool publish_agg = true) {
  SklOp op;
  const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
  __shared__ int s_p;
  __shared__ SKL_T s_wv[SKL_NW];
  __shared__ SKL_T s_acc;
  if (tile == 0) {
    if (tid == 0) {
      const SKL_T agg = *s_agg;
      if (ncarry > 0) {  // multi-GPU carry-in: totals of the preceding devices
        SKL_T c = carry[0];
        for (int i = 1; i < ncarry; ++i) c = op(c, carry[i]);
        skl_publish(flags, aggs, incls, 0, epoch, 2u, op(c, agg));
        *s_excl = c;
        *s_has = 1;
      } else {
        skl_publish(flags, aggs, incls, 0, epoch, 2u, agg);
        *s_has = 0;
      }
    }
    return;
  }
  if (tid == 0 && publish_agg) skl_publish(flags, aggs, incls, tile, epoch, 1u, *s_agg);
  bool have = false;  // thread 0 only
  long base = (long)tile - 1;
  // each thread watches SKL_LBW consecutive predecessors (distances tid*W ..
  // tid*W + W-1), their loads issued together: one round trip covers
  // SKL_BLOCK x SKL_LBW tiles (>= the tiles in flight, so usually one round)
  constexpr int W = SKL_LBW;
  while (true) {
    SKL_T val[W];
    unsigned st[W];
#pragma unroll
    for (int r = 0; r < W; ++r) st[r] = 0u;
    for (bool pending = true; pending;) {
      pending = false;
#pragma unroll
      for (int r = 0; r < W; ++r) {
        const long j = base - (long)(tid * W + r);
        if (j >= 0 && st[r] == 0u) {
          st[r] = skl_status_try(flags, aggs, incls, j, epoch, &val[r]);
          pending |= st[r] == 0u;
        }
      }
    }
    int myp = W * SKL_BLOCK;
#pragma unroll
    for (int r = W - 1; r >= 0; --r)
      if (st[r] == 2u) myp = tid * W + r;  // nearest prefix among mine
    if (tid == 0) s_p = W * SKL_BLOCK;
    __syncthreads();
    if (myp < W * SKL_BLOCK) atomicMin(&s_p, myp);
    __syncthreads();
    const int pfound = s_p;  // distance of the nearest inclusive prefix
    const int plim = pfound < W * SKL_BLOCK ? pfound : W * SKL_BLOCK - 1;
    // thread-local fold of my distances <= plim, the larger distance on the left
    SKL_T v;
    bool hv = false;
#pragma unroll
    for (int r = W - 1; r >= 0; --r) {
      const int dist = tid * W + r;
      if (dist <= plim && base - (long)dist >= 0) {
        v = hv ? op(v, val[r]) : val[r];
        hv = true;
      }
    }
    const int p = plim / W;  // threads 0..p contribute
    // fold threads p..0 (a higher thread is an earlier tile: the left operand)
    const int wp = p - warp * 32;  // last contributing lane of this warp
#pragma unroll
    for (int s = 1; s < 32; s <<= 1) {
      SKL_T o = skl_shfl_down(v, s);
      if (lane + s <= wp) v = op(o, v);
    }
    if (lane == 0 && wp >= 0) s_wv[warp] = v;
    __syncthreads();
    if (tid == 0) {
      SKL_T w = s_wv[p / 32];
      for (int k = p / 32 - 1; k >= 0; --k) w = op(w, s_wv[k]);
      s_acc = have ? op(w, s_acc) : w;
      have = true;
    }
    if (pfound < W * SKL_BLOCK) break;
    base -= W * SKL_BLOCK;
    __syncthreads();  // s_p / s_wv are reused by the next round
  }
  if (tid == 0) {
    skl_publish(flags, aggs, incls, tile, epoch, 2u, op(s_acc, *s_agg));
    *s_excl = s_acc;
    *s_has = 1;
  }
}

// Warp-wide look-back (called by warp 0 only): 32 predecessors per round trip,
// no block barriers inside the spin.
__device__ __forceinline__ void skl_lookback_warp(unsigned tile, unsigned* flags, SKL_T* aggs,
                                                  SKL_T* incls, unsigned epoch, const SKL_T* carry,
                                                  int ncarry, const SKL_T* s_agg, SKL_T* s_excl,
                                                  int* s_has) {
  SklOp op;
  const int lane = threadIdx.x & 31;
  if (tile == 0) {
    if (lane == 0) {
      const SKL_T agg = *s_agg;
      if (ncarry > 0) {
        SKL_T c = carry[0];
        for (int i = 1; i < ncarry; ++i) c = op(c, carry[i]);
        skl_publish(flags, aggs, incls, 0, epoch, 2u, op(c, agg));
        *s_excl = c;
        *s_has = 1;
      } else {
        skl_publish(flags, aggs, incls, 0, epoch, 2u, agg);
        *s_has = 0;
      }
    }
    return;
  }
  if (lane == 0) skl_publish(flags, aggs, incls, tile, epoch, 1u, *s_agg);
  bool have = false;
  SKL_T acc;
  long base = (long)tile - 1;
  while (true) {
    const long j = base - lane;
    SKL_T v;
    unsigned st = 0;
    if (j >= 0) st = skl_status(flags, aggs, incls, j, epoch, &v);
    const unsigned pm = __ballot_sync(SKL_FULL, st == 2u);
    const int p = pm ? __ffs(pm) - 1 : 31;
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
    skl_publish(flags, aggs, incls, tile, epoch, 2u, op(acc, *s_agg));
    *s_excl = acc;
    *s_has = 1;
  }
}

// Shared body: items[] holds this thread's (blocked) elements, cnt of them valid.
// On return items[k] holds the inclusive scan value of element t*ITEMS+k.
// LOOKBACK = false: the tile's exclusive prefix is given (pre_has, pre) instead of
// looked back, and the tile aggregate is returned in *agg_out (all threads).
template <int ITEMS, bool LOOKBACK = true>
__device__ __forceinline__ void skl_scan_tile(SKL_T (&items)[ITEMS], int cnt, int nthr_valid,
                                              unsigned tile, unsigned* flags, SKL_T* aggs, SKL_T* incls,
                                              unsigned epoch, const SKL_T* carry, int ncarry,
                                              bool pre_has = false, const SKL_T* pre_in = nullptr,
                                              SKL_T* agg_out = nullptr, int* pre_has_out = nullptr,
                                              SKL_T* pre_out = nullptr) {
  SklOp op;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  // 1. sequential inclusive scan inside the thread
  SKL_T v = items[0];
#pragma unroll
  for (int k = 1; k < ITEMS; ++k)
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
  // 4. look-back for the tile prefix (whole block: SKL_BLOCK predecessors per round trip)
  if (!LOOKBACK) {
    if (threadIdx.x == 0) {
      s_has = pre_has;
      if (pre_has) s_excl = *pre_in;
    }
  } else {
#if SKL_SCAN_VARIANT == 1 || SKL_SCAN_VARIANT == 7
    // measurement variant only (skl_set_option "scan_variant" 1): no look-back,
    // i.e. per-tile scans - the load/scan/store pipeline's own ceiling
    if (threadIdx.x == 0) s_has = 0;
#elif SKL_SCAN_VARIANT == 2
    if ((threadIdx.x >> 5) == 0)
      skl_lookback_warp(tile, flags, aggs, incls, epoch, carry, ncarry, &s_agg, &s_excl, &s_has);
#else
    skl_lookback_block(tile, flags, aggs, incls, epoch, carry, ncarry, &s_agg, &s_excl, &s_has);
#endif
  }
  __syncthreads();
  if (agg_out) *agg_out = s_agg;
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
  if (pre_has_out) {  // the caller applies the prefix itself
    *pre_has_out = hp;
    if (hp) *pre_out = pre;
    return;
  }
  if (hp) {
#pragma unroll
    for (int k = 0; k < ITEMS; ++k)
      if (k < cnt) items[k] = op(pre, items[k]);
  }
}

#if SKL_CH > 0
// Vector path (sizeof(T) divides 16, in/out 16-byte aligned): chained scan over
// L2-resident chunks.  A tile-granular look-back couples the blocks in
// lock-step rounds of one 32 KB tile each, and the look-back latency per round
// then dominates (measured: 2.3-2.5 TB/s; 6.5 TB/s without look-back).  Here a
// persistent block takes chunks c = b, b + grid, ... of SKL_SUB tiles:
//   pass 1  order-preserving fold of the chunk straight from HBM (registers,
//           16-byte loads, SKL_RU warp-tiles in flight per warp) -> publish the
//           chunk aggregate, look back (one round trip covers SKL_BLOCK chunks);
//   pass 2  re-read the chunk (an L2 hit: grid x chunk bytes << 126 MB), scan
//           its tiles in order from shared memory (cp.async double buffer, XOR
//           swizzle) with a running prefix, stream the result out.
// HBM traffic stays 8 B per 4-byte element; the look-back rounds shrink SKL_SUB x.
#define SKL_EPC (16 / (int)sizeof(SKL_T))  // elements per 16-byte chunk
#ifndef SKL_SUB
#define SKL_SUB 4
#endif
#define SKL_CHUNK ((skl_u64)SKL_TILE * SKL_SUB)
__device__ __forceinline__ void skl_cp16(void* smem, const void* g) {
  const unsigned s = (unsigned)__cvta_generic_to_shared(smem);
  asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" ::"r"(s), "l"(g) : "memory");
}
__device__ __forceinline__ void skl_cp_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
__device__ __forceinline__ void skl_cp_wait1() { asm volatile("cp.async.wait_group 1;" ::: "memory"); }

// stage the tile [tlo, tlo + nvalid) into sm: full 16-byte chunks asynchronously,
// a ragged tail synchronously
__device__ __forceinline__ void skl_scan_issue(const SKL_T* __restrict__ in, skl_u64 tlo, int nvalid,
                                               uint4* sm) {
  const char* gin = (const char*)(in + tlo);
  if (nvalid == SKL_TILE) {
#pragma unroll
    for (int i = 0; i < SKL_CH; ++i) {
      const unsigned c = i * SKL_BLOCK + threadIdx.x;
      skl_cp16(&sm[skl_swz(c)], gin + 16 * (skl_u64)c);
    }
  } else {
    const int nfull = nvalid / SKL_EPC;
    for (int c = threadIdx.x; c < nfull; c += SKL_BLOCK) skl_cp16(&sm[skl_swz(c)], gin + 16 * (skl_u64)c);
    for (int e = nfull * SKL_EPC + threadIdx.x; e < nvalid; e += SKL_BLOCK)
      *((SKL_T*)&sm[skl_swz(e / SKL_EPC)] + (e % SKL_EPC)) = in[tlo + e];
  }
}

// Ordered fold of [lo, hi) by one warp: warp-tiles of 32 lanes x SKL_EPC
// elements (one 16-byte load per lane), SKL_RU warp-tiles in flight.
__device__ __forceinline__ void skl_warp_range_fold(const SKL_T* __restrict__ in, skl_u64 lo, skl_u64 hi,
                                                    bool& has, SKL_T& acc) {
  SklOp op;
  const int lane = threadIdx.x & 31;
  const skl_u64 wt = 32 * SKL_EPC;
  for (skl_u64 t = lo; t < hi; t += wt * SKL_RU) {
    SKL_T x[SKL_RU][SKL_EPC];
    int cnt[SKL_RU];
#pragma unroll
    for (int u = 0; u < SKL_RU; ++u) {
      const skl_u64 e = t + u * wt + (skl_u64)lane * SKL_EPC;
      cnt[u] = e >= hi ? 0 : (hi - e >= (skl_u64)SKL_EPC ? SKL_EPC : (int)(hi - e));
      if (cnt[u] == SKL_EPC) {
        SklChunk<SKL_T, SKL_EPC> ch;
        ch.q[0] = skl_ld16(in + e);
#pragma unroll
        for (int k = 0; k < SKL_EPC; ++k) x[u][k] = ch.e[k];
      } else {
#pragma unroll
        for (int k = 0; k < SKL_EPC; ++k)
          if (k < cnt[u]) x[u][k] = in[e + k];
      }
    }
#pragma unroll
    for (int u = 0; u < SKL_RU; ++u) {
      const skl_u64 tl = t + u * wt;
      if (tl >= hi) break;
      SKL_T v = x[u][0];
#pragma unroll
      for (int k = 1; k < SKL_EPC; ++k)
        if (k < cnt[u]) v = op(v, x[u][k]);
      const skl_u64 rem = hi - tl;
      const int nv = rem >= wt ? 32 : (int)((rem + SKL_EPC - 1) / SKL_EPC);
      v = skl_warp_fold(v, nv, op);
      v = skl_shfl(v, 0);
      acc = has ? op(acc, v) : v;
      has = true;
    }
  }
}

// ---- persistent, 3-stage software pipeline (SKL_SCAN_VARIANT 4) -------------
// Block b owns tiles t_k = b + k * grid.  Iteration k:
//   issue the load of t_{k+2} (cp.async, stage (k+2) % 3)
//   look back for t_k            (its aggregate was published one iteration ago,
//                                 so predecessors in the same round are ready)
//   apply the tile prefix to t_k's locally scanned values, stream them out
//   local scan of t_{k+1} (landed meanwhile), publish its aggregate
// so the look-back latency overlaps loads already in flight instead of stalling
// the memory pipeline (the per-tile kernel's top stalls were barriers and the
// look-back spin; the same tile pipeline without look-back runs at copy speed).
#ifndef SKL_MINB_P
#define SKL_MINB_P 1
#endif
__device__ __forceinline__ int skl_nvalid(skl_u64 n, unsigned t) {
  const skl_u64 tlo = (skl_u64)t * SKL_TILE;
  return n - tlo >= (skl_u64)SKL_TILE ? SKL_TILE : (int)(n - tlo);
}

// local (within-tile) inclusive scan of the tile in stage sm, written back in
// place; returns the tile aggregate (all threads)
__device__ __forceinline__ SKL_T skl_tile_local(uint4* sm, int nvalid) {
  SklChunk<SKL_T, SKL_ITEMS> my;
#pragma unroll
  for (int q = 0; q < SKL_CH; ++q) my.q[q] = sm[skl_swz(threadIdx.x * SKL_CH + q)];
  SKL_T items[SKL_ITEMS];
#pragma unroll
  for (int q = 0; q < SKL_ITEMS; ++q) items[q] = my.e[q];
  const int first = threadIdx.x * SKL_ITEMS;
  const int cnt = nvalid - first >= SKL_ITEMS ? SKL_ITEMS : (nvalid - first > 0 ? nvalid - first : 0);
  const int nthr = (nvalid + SKL_ITEMS - 1) / SKL_ITEMS;
  SKL_T agg;
  skl_scan_tile<SKL_ITEMS, false>(items, cnt, nthr, 0, nullptr, nullptr, nullptr, 0, nullptr, 0, false,
                                  nullptr, &agg);
#pragma unroll
  for (int q = 0; q < SKL_ITEMS; ++q) my.e[q] = items[q];
#pragma unroll
  for (int q = 0; q < SKL_CH; ++q) sm[skl_swz(threadIdx.x * SKL_CH + q)] = my.q[q];
  return agg;
}

extern "C" __global__ void __launch_bounds__(SKL_BLOCK, SKL_MINB_P)
skl_scan_pipe(const SKL_T* __restrict__ in, SKL_T* __restrict__ out, skl_u64 n, unsigned* flags,
              SKL_T* aggs, SKL_T* incls, unsigned epoch, const SKL_T* carry, int ncarry) {
  extern __shared__ uint4 skl_dyn[];
  __shared__ SKL_T p_agg[3];
  __shared__ SKL_T p_excl;
  __shared__ int p_has;
  SklOp op;
  const unsigned ntiles = (unsigned)((n + SKL_TILE - 1) / SKL_TILE);
  const unsigned G = gridDim.x;
  const unsigned t0 = blockIdx.x;
  if (t0 >= ntiles) return;
#define SKL_STAGE(k) (skl_dyn + ((k) % 3u) * (SKL_BLOCK * SKL_CH))
  skl_scan_issue(in, (skl_u64)t0 * SKL_TILE, skl_nvalid(n, t0), SKL_STAGE(0u));
  skl_cp_commit();
  if (t0 + G < ntiles) skl_scan_issue(in, (skl_u64)(t0 + G) * SKL_TILE, skl_nvalid(n, t0 + G), SKL_STAGE(1u));
  skl_cp_commit();
  skl_cp_wait1();
  __syncthreads();
  {
    const SKL_T agg = skl_tile_local(SKL_STAGE(0u), skl_nvalid(n, t0));
    if (threadIdx.x == 0) {
      p_agg[0] = agg;
      if (t0 != 0) skl_publish(flags, aggs, incls, t0, epoch, 1u, agg);  // tile 0 publishes P
    }
  }
  __syncthreads();
  for (unsigned k = 0;; ++k) {
    const unsigned t = t0 + k * G;
    if (t >= ntiles) break;
    const unsigned t1 = t + G, t2 = t + 2 * G;
    if (t2 < ntiles) skl_scan_issue(in, (skl_u64)t2 * SKL_TILE, skl_nvalid(n, t2), SKL_STAGE(k + 2));
    skl_cp_commit();
    // ---- look-back for t (aggregate already public)
#if SKL_SCAN_VARIANT == 5
    if (threadIdx.x == 0) p_has = 0;  // measurement only: no look-back
#else
    skl_lookback_block(t, flags, aggs, incls, epoch, carry, ncarry, &p_agg[k % 3], &p_excl, &p_has, false);
#endif
    __syncthreads();
    // ---- apply the tile prefix, stream out
    {
      uint4* sm = SKL_STAGE(k);
      const int nvalid = skl_nvalid(n, t);
      const bool has = p_has != 0;
      const SKL_T pre = p_excl;
      const skl_u64 tlo = (skl_u64)t * SKL_TILE;
      char* gout = (char*)(out + tlo);
      if (nvalid == SKL_TILE) {
#pragma unroll
        for (int i = 0; i < SKL_CH; ++i) {
          const unsigned c = i * SKL_BLOCK + threadIdx.x;
          SklChunk<SKL_T, SKL_EPC> ch;
          ch.q[0] = sm[skl_swz(c)];
          if (has) {
#pragma unroll
            for (int e = 0; e < SKL_EPC; ++e) ch.e[e] = op(pre, ch.e[e]);
          }
          skl_st16(gout + 16 * (skl_u64)c, ch.q[0]);
        }
      } else {
        for (int e = threadIdx.x; e < nvalid; e += SKL_BLOCK) {
          SKL_T v = *((const SKL_T*)&sm[skl_swz(e / SKL_EPC)] + (e % SKL_EPC));
          out[tlo + e] = has ? op(pre, v) : v;
        }
      }
    }
    // ---- local scan of t1 (landed while this tile looked back)
    if (t1 < ntiles) {
      skl_cp_wait1();
      __syncthreads();  // t1 visible; every thread is past this tile's apply
      const SKL_T agg = skl_tile_local(SKL_STAGE(k + 1), skl_nvalid(n, t1));
      if (threadIdx.x == 0) {
        p_agg[(k + 1) % 3] = agg;
        skl_publish(flags, aggs, incls, t1, epoch, 1u, agg);
      }
    }
    __syncthreads();  // stage k is refilled by the next iteration's prefetch
  }
#undef SKL_STAGE
}

// One block per tile (tile = blockIdx.x; blocks start in index order), tile
// look-back (SKL_SCAN_VARIANT 2: warp-wide window; else block-wide).
#ifndef SKL_MINB
#define SKL_MINB 1
#endif
extern "C" __global__ void __launch_bounds__(SKL_BLOCK, SKL_MINB)
skl_scan_pt(const SKL_T* __restrict__ in, SKL_T* __restrict__ out, skl_u64 n, unsigned* flags,
            SKL_T* aggs, SKL_T* incls, unsigned epoch, const SKL_T* carry, int ncarry) {
  extern __shared__ uint4 skl_dyn[];
  uint4* sm = skl_dyn;
  const unsigned t = blockIdx.x;
  const skl_u64 tlo = (skl_u64)t * SKL_TILE;
  const int nvalid = n - tlo >= (skl_u64)SKL_TILE ? SKL_TILE : (int)(n - tlo);
  skl_scan_issue(in, tlo, nvalid, sm);
  skl_cp_commit();
  asm volatile("cp.async.wait_group 0;" ::: "memory");
  __syncthreads();
  SklChunk<SKL_T, SKL_ITEMS> my;
#pragma unroll
  for (int q = 0; q < SKL_CH; ++q) my.q[q] = sm[skl_swz(threadIdx.x * SKL_CH + q)];
  SKL_T items[SKL_ITEMS];
#pragma unroll
  for (int q = 0; q < SKL_ITEMS; ++q) items[q] = my.e[q];
  const int first = threadIdx.x * SKL_ITEMS;
  const int cnt = nvalid - first >= SKL_ITEMS ? SKL_ITEMS : (nvalid - first > 0 ? nvalid - first : 0);
  const int nthr = (nvalid + SKL_ITEMS - 1) / SKL_ITEMS;
  skl_scan_tile<SKL_ITEMS, true>(items, cnt, nthr, t, flags, aggs, incls, epoch, carry, ncarry);
#pragma unroll
  for (int q = 0; q < SKL_ITEMS; ++q) my.e[q] = items[q];
#pragma unroll
  for (int q = 0; q < SKL_CH; ++q) sm[skl_swz(threadIdx.x * SKL_CH + q)] = my.q[q];
  __syncthreads();
  char* gout = (char*)(out + tlo);
  if (nvalid == SKL_TILE) {
#pragma unroll
    for (int i = 0; i < SKL_CH; ++i) {
      const unsigned cc = i * SKL_BLOCK + threadIdx.x;
      skl_st16(gout + 16 * (skl_u64)cc, sm[skl_swz(cc)]);
    }
  } else {
    for (int e = threadIdx.x; e < nvalid; e += SKL_BLOCK)
      out[tlo + e] = *((const SKL_T*)&sm[skl_swz(e / SKL_EPC)] + (e % SKL_EPC));
  }
}

// Low-register per-tile variant (SKL_SCAN_VARIANT 6): the tile stays in shared
// memory; a thread folds its SKL_ITEMS elements to one total (16-byte reads),
// the block scans the totals and looks back, then the thread re-reads its
// elements and writes pre (+) x0, (pre (+) x0) (+) x1, ... in place.  No item
// array lives in registers, so more tiles (SKL_MINB) fit per SM: the look-back
// latency of one tile is hidden behind the loads of the others.
extern "C" __global__ void __launch_bounds__(SKL_BLOCK, SKL_MINB)
skl_scan_lr(const SKL_T* __restrict__ in, SKL_T* __restrict__ out, skl_u64 n, unsigned* flags,
            SKL_T* aggs, SKL_T* incls, unsigned epoch, const SKL_T* carry, int ncarry) {
  extern __shared__ uint4 skl_dyn[];
  uint4* sm = skl_dyn;
  SklOp op;
  const unsigned t = blockIdx.x;
  const skl_u64 tlo = (skl_u64)t * SKL_TILE;
  const int nvalid = n - tlo >= (skl_u64)SKL_TILE ? SKL_TILE : (int)(n - tlo);
  skl_scan_issue(in, tlo, nvalid, sm);
  skl_cp_commit();
  asm volatile("cp.async.wait_group 0;" ::: "memory");
  __syncthreads();
  const int first = threadIdx.x * SKL_ITEMS;
  const int cnt = nvalid - first >= SKL_ITEMS ? SKL_ITEMS : (nvalid - first > 0 ? nvalid - first : 0);
  const int nthr = (nvalid + SKL_ITEMS - 1) / SKL_ITEMS;
#define SKL_LR_ELT(k) (*((SKL_T*)&sm[skl_swz((unsigned)(first + (k)) / SKL_EPC)] + ((first + (k)) % SKL_EPC)))
  SKL_T tot[1];
  if (cnt == SKL_ITEMS) {
    SklChunk<SKL_T, SKL_EPC> c0;
    c0.q[0] = sm[skl_swz(threadIdx.x * SKL_CH)];
    tot[0] = c0.e[0];
#pragma unroll
    for (int e = 1; e < SKL_EPC; ++e) tot[0] = op(tot[0], c0.e[e]);
#pragma unroll
    for (int q = 1; q < SKL_CH; ++q) {
      SklChunk<SKL_T, SKL_EPC> c;
      c.q[0] = sm[skl_swz(threadIdx.x * SKL_CH + q)];
#pragma unroll
      for (int e = 0; e < SKL_EPC; ++e) tot[0] = op(tot[0], c.e[e]);
    }
  } else if (cnt > 0) {
    tot[0] = SKL_LR_ELT(0);
    for (int k = 1; k < cnt; ++k) tot[0] = op(tot[0], SKL_LR_ELT(k));
  }
  int hp = 0;
  SKL_T pre;
  skl_scan_tile<1, true>(tot, cnt > 0 ? 1 : 0, nthr, t, flags, aggs, incls, epoch, carry, ncarry, false,
                         nullptr, nullptr, &hp, &pre);
  if (cnt == SKL_ITEMS) {
#pragma unroll
    for (int q = 0; q < SKL_CH; ++q) {
      SklChunk<SKL_T, SKL_EPC> c;
      c.q[0] = sm[skl_swz(threadIdx.x * SKL_CH + q)];
#pragma unroll
      for (int e = 0; e < SKL_EPC; ++e) {
        if (q == 0 && e == 0) {
          if (hp) c.e[0] = op(pre, c.e[0]);
        } else {
          c.e[e] = op(pre, c.e[e]);
        }
        pre = c.e[e];
      }
      sm[skl_swz(threadIdx.x * SKL_CH + q)] = c.q[0];
    }
  } else if (cnt > 0) {
    for (int k = 0; k < cnt; ++k) {
      SKL_T v = SKL_LR_ELT(k);
      if (k > 0 || hp) v = op(pre, v);
      SKL_LR_ELT(k) = v;
      pre = v;
    }
  }
#undef SKL_LR_ELT
  __syncthreads();
  char* gout = (char*)(out + tlo);
  if (nvalid == SKL_TILE) {
#pragma unroll
    for (int i = 0; i < SKL_CH; ++i) {
      const unsigned cc = i * SKL_BLOCK + threadIdx.x;
      skl_st16(gout + 16 * (skl_u64)cc, sm[skl_swz(cc)]);
    }
  } else {
    for (int e = threadIdx.x; e < nvalid; e += SKL_BLOCK)
      out[tlo + e] = *((const SKL_T*)&sm[skl_swz(e / SKL_EPC)] + (e % SKL_EPC));
  }
}

extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_scan_vec(const SKL_T* __restrict__ in, SKL_T* __restrict__ out, skl_u64 n, unsigned* flags,
             SKL_T* aggs, SKL_T* incls, unsigned epoch, const SKL_T* carry, int ncarry) {
  extern __shared__ uint4 skl_dyn[];
  SklOp op;
  const int warp = threadIdx.x >> 5;
  __shared__ SKL_T c_wv[SKL_NW];
  __shared__ int c_wh[SKL_NW];
  __shared__ SKL_T c_agg, c_excl;
  __shared__ int c_has;
  const unsigned nchunks = (unsigned)((n + SKL_CHUNK - 1) / SKL_CHUNK);
  for (unsigned c = blockIdx.x; c < nchunks; c += gridDim.x) {
    const skl_u64 clo = (skl_u64)c * SKL_CHUNK;
    const skl_u64 chi = n - clo > SKL_CHUNK ? clo + SKL_CHUNK : n;
    // ---- pass 1: chunk aggregate (warps own consecutive equal slices)
    {
      const skl_u64 wlen = SKL_CHUNK / SKL_NW;
      const skl_u64 wlo = clo + (skl_u64)warp * wlen;
      const skl_u64 whi = wlo + wlen < chi ? wlo + wlen : chi;
      bool has = false;
      SKL_T acc;
      if (wlo < chi) skl_warp_range_fold(in, wlo, whi, has, acc);
      if ((threadIdx.x & 31) == 0) {
        c_wh[warp] = has;
        if (has) c_wv[warp] = acc;
      }
      __syncthreads();
      if (threadIdx.x == 0) {
        SKL_T a = c_wv[0];
        for (int w = 1; w < SKL_NW; ++w)
          if (c_wh[w]) a = op(a, c_wv[w]);
        c_agg = a;
      }
      __syncthreads();
    }
#if SKL_SCAN_VARIANT == 1
    if (threadIdx.x == 0) c_has = 0;
#else
    skl_lookback_block(c, flags, aggs, incls, epoch, carry, ncarry, &c_agg, &c_excl, &c_has);
#endif
    __syncthreads();
    // ---- pass 2: tiles of the chunk in order, running prefix, from L2
    bool run_has = c_has != 0;
    SKL_T run;
    if (run_has) run = c_excl;
    const unsigned ntile = (unsigned)((chi - clo + SKL_TILE - 1) / SKL_TILE);
    skl_scan_issue(in, clo, chi - clo >= (skl_u64)SKL_TILE ? SKL_TILE : (int)(chi - clo), skl_dyn);
    skl_cp_commit();
    for (unsigned k = 0; k < ntile; ++k) {
      uint4* sm = skl_dyn + (k & 1) * (SKL_BLOCK * SKL_CH);
      const skl_u64 tlo = clo + (skl_u64)k * SKL_TILE;
      const int nvalid = chi - tlo >= (skl_u64)SKL_TILE ? SKL_TILE : (int)(chi - tlo);
      if (k + 1 < ntile) {
        const skl_u64 nlo = tlo + SKL_TILE;
        skl_scan_issue(in, nlo, chi - nlo >= (skl_u64)SKL_TILE ? SKL_TILE : (int)(chi - nlo),
                       skl_dyn + ((k + 1) & 1) * (SKL_BLOCK * SKL_CH));
      }
      skl_cp_commit();
      skl_cp_wait1();
      __syncthreads();
      SklChunk<SKL_T, SKL_ITEMS> my;
#pragma unroll
      for (int q = 0; q < SKL_CH; ++q) my.q[q] = sm[skl_swz(threadIdx.x * SKL_CH + q)];
      SKL_T items[SKL_ITEMS];
#pragma unroll
      for (int q = 0; q < SKL_ITEMS; ++q) items[q] = my.e[q];
      const int first = threadIdx.x * SKL_ITEMS;
      const int cnt = nvalid - first >= SKL_ITEMS ? SKL_ITEMS : (nvalid - first > 0 ? nvalid - first : 0);
      const int nthr = (nvalid + SKL_ITEMS - 1) / SKL_ITEMS;
      SKL_T tagg;
      skl_scan_tile<SKL_ITEMS, false>(items, cnt, nthr, 0, flags, aggs, incls, epoch, carry, ncarry,
                                      run_has, &run, &tagg);
      run = run_has ? op(run, tagg) : tagg;
      run_has = true;
#pragma unroll
      for (int q = 0; q < SKL_ITEMS; ++q) my.e[q] = items[q];
#pragma unroll
      for (int q = 0; q < SKL_CH; ++q) sm[skl_swz(threadIdx.x * SKL_CH + q)] = my.q[q];
      __syncthreads();
      char* gout = (char*)(out + tlo);
      if (nvalid == SKL_TILE) {
#pragma unroll
        for (int i = 0; i < SKL_CH; ++i) {
          const unsigned cc = i * SKL_BLOCK + threadIdx.x;
          skl_st16(gout + 16 * (skl_u64)cc, sm[skl_swz(cc)]);
        }
      } else {
        for (int e = threadIdx.x; e < nvalid; e += SKL_BLOCK)
          out[tlo + e] = *((const SKL_T*)&sm[skl_swz(e / SKL_EPC)] + (e % SKL_EPC));
      }
      __syncthreads();  // this stage is refilled by the next prefetch
    }
  }
}
#endif

// Generic path: any element size / alignment (blocked layout through smem), one
// block per tile of SKL_BLOCK x SKL_SC_ITEMS elements.
#define SKL_SC_ITEMS 8
#define SKL_SC_TILE (SKL_BLOCK * SKL_SC_ITEMS)
extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_scan_sc(const SKL_T* __restrict__ in, SKL_T* __restrict__ out, skl_u64 n, unsigned* flags,
            SKL_T* aggs, SKL_T* incls, unsigned epoch, const SKL_T* carry, int ncarry) {
  __shared__ __align__(16) unsigned char sm_raw[SKL_SC_TILE * sizeof(SKL_T)];
  SKL_T* sm_u = (SKL_T*)sm_raw;
  const skl_u64 tlo = (skl_u64)blockIdx.x * SKL_SC_TILE;
  const int nvalid = n - tlo >= (skl_u64)SKL_SC_TILE ? SKL_SC_TILE : (int)(n - tlo);
  for (int e = threadIdx.x; e < nvalid; e += SKL_BLOCK) sm_u[e] = in[tlo + e];
  __syncthreads();
  SKL_T items[SKL_SC_ITEMS];
  const int first = threadIdx.x * SKL_SC_ITEMS;
#pragma unroll
  for (int k = 0; k < SKL_SC_ITEMS; ++k)
    if (first + k < nvalid) items[k] = sm_u[first + k];
  const int cnt = nvalid - first >= SKL_SC_ITEMS ? SKL_SC_ITEMS : (nvalid - first > 0 ? nvalid - first : 0);
  const int nthr = (nvalid + SKL_SC_ITEMS - 1) / SKL_SC_ITEMS;
  skl_scan_tile<SKL_SC_ITEMS>(items, cnt, nthr, blockIdx.x, flags, aggs, incls, epoch, carry, ncarry);
  __syncthreads();
#pragma unroll
  for (int k = 0; k < SKL_SC_ITEMS; ++k)
    if (k < cnt) sm_u[first + k] = items[k];
  __syncthreads();
  for (int e = threadIdx.x; e < nvalid; e += SKL_BLOCK) out[tlo + e] = sm_u[e];
}
