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

// Element loaders: the plain Reduce reads its input; the fused form (lazy
// Zip/Map -> Reduce) computes each element from the Zip's inputs
// on the fly, so the intermediate vector never exists (8 instead of 16 bytes per
// element for the dot product of Listing 1.1).
struct SklLoadPlain {
  const SKL_T* __restrict__ in;
  template <int RVEC>
  __device__ __forceinline__ void load(skl_u64 e, int cnt, SKL_T (&x)[RVEC]) const {
    if (RVEC > 1 && cnt == RVEC) {
      SklChunk<SKL_T, RVEC> ch;
      ch.q[0] = skl_ld16(in + e);
#pragma unroll
      for (int k = 0; k < RVEC; ++k) x[k] = ch.e[k];
    } else {
#pragma unroll
      for (int k = 0; k < RVEC; ++k)
        if (k < cnt) x[k] = in[e + k];
    }
  }
};
#if SKL_FUSED
struct SklLoadZip {
  const SKL_ZL* __restrict__ l;
  const SKL_ZR* __restrict__ r;
  __device__ __forceinline__ SKL_T f(const SKL_ZL& a, const SKL_ZR& b) const {
#if SKL_ZMAP
    (void)b;
    return SKL_ZFUNC(a);
#else
    return SKL_ZFUNC(a, b);
#endif
  }
  template <int RVEC>
  __device__ __forceinline__ void load(skl_u64 e, int cnt, SKL_T (&x)[RVEC]) const {
    if (RVEC > 1 && cnt == RVEC) {
      SklChunk<SKL_ZL, RVEC> a;
      a.q[0] = skl_ld16(l + e);
#if SKL_ZMAP
#pragma unroll
      for (int k = 0; k < RVEC; ++k) x[k] = f(a.e[k], a.e[k]);
#else
      SklChunk<SKL_ZR, RVEC> b;
      b.q[0] = skl_ld16(r + e);
#pragma unroll
      for (int k = 0; k < RVEC; ++k) x[k] = f(a.e[k], b.e[k]);
#endif
    } else {
#pragma unroll
      for (int k = 0; k < RVEC; ++k)
        if (k < cnt) {
#if SKL_ZMAP
          x[k] = f(l[e + k], l[e + k]);
#else
          x[k] = f(l[e + k], r[e + k]);
#endif
        }
    }
  }
};
#endif

template <int RVEC, class Loader>
__device__ __forceinline__ void skl_reduce_body(const Loader& ld, skl_u64 n, skl_u64 wseg,
                                                SKL_T* partials, unsigned* counter, SKL_T* result) {
  SklOp op;
  // a warp-tile is 32 lanes x RVEC elements of THIS instantiation (the scalar
  // kernel, RVEC = 1, serves unaligned views)
  constexpr skl_u64 RT = 32 * RVEC;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const skl_u64 w = (skl_u64)blockIdx.x * SKL_NW + warp;
  const skl_u64 lo = w * wseg;
  const skl_u64 hi = lo + wseg < n ? lo + wseg : n;
  bool has = false;
  SKL_T acc;
  skl_u64 t = lo;
  // fast path: SKL_RU full warp-tiles, no per-tile branches, so all loads of the
  // iteration are issued before the first use (memory-level parallelism)
  for (; t + RT * SKL_RU <= hi; t += RT * SKL_RU) {
    SKL_T x[SKL_RU][RVEC];
#pragma unroll
    for (int u = 0; u < SKL_RU; ++u)
      ld.template load<RVEC>(t + (skl_u64)u * RT + (skl_u64)lane * RVEC, RVEC, x[u]);
#pragma unroll
    for (int u = 0; u < SKL_RU; ++u) {
      SKL_T v = x[u][0];
#pragma unroll
      for (int k = 1; k < RVEC; ++k) v = op(v, x[u][k]);
      v = skl_warp_fold(v, 32, op);
      v = skl_shfl(v, 0);
      acc = has ? op(acc, v) : v;
      has = true;
    }
  }
  // ragged end of the segment
  for (; t < hi; t += RT * SKL_RU) {
    SKL_T x[SKL_RU][RVEC];
    int cnt[SKL_RU];
#pragma unroll
    for (int u = 0; u < SKL_RU; ++u) {
      const skl_u64 e = t + (skl_u64)u * RT + (skl_u64)lane * RVEC;
      cnt[u] = e >= hi ? 0 : (hi - e >= (skl_u64)RVEC ? RVEC : (int)(hi - e));
      ld.template load<RVEC>(e, cnt[u], x[u]);
    }
#pragma unroll
    for (int u = 0; u < SKL_RU; ++u) {
      const skl_u64 tl = t + (skl_u64)u * RT;
      if (tl >= hi) break;
      SKL_T v = x[u][0];
#pragma unroll
      for (int k = 1; k < RVEC; ++k)
        if (k < cnt[u]) v = op(v, x[u][k]);
      const skl_u64 rem = hi - tl;
      const int nv = rem >= RT ? 32 : (int)((rem + RVEC - 1) / RVEC);
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
      // release: the partial is visible before the ticket (no separate fence,
      // one L2 round trip on the critical path instead of two)
      unsigned ticket;
      asm volatile("atom.add.acq_rel.gpu.global.u32 %0, [%1], 1;" : "=r"(ticket) : "l"(counter) : "memory");
      s_last = (ticket == gridDim.x - 1);
    }
  }
  if (gridDim.x == 1) return;
  __syncthreads();
  if (!s_last) return;
  // last block: fold the block partials in block order, every warp folding one
  // contiguous slice (one L2 round trip per 32 x SKL_NW partials), then the warp
  // results in warp order
  __threadfence();
  const unsigned per = (gridDim.x + SKL_NW - 1) / SKL_NW;
  const unsigned wlo = warp * per;
  const unsigned whi = wlo + per < gridDim.x ? wlo + per : gridDim.x;
  bool h2 = false;
  SKL_T a2;
  for (unsigned b0 = wlo; b0 < whi; b0 += 32) {
    const unsigned nb = whi - b0 < 32 ? whi - b0 : 32;
    SKL_T v;
    if ((unsigned)lane < nb) v = skl_ldcg(partials + b0 + lane);
    v = skl_warp_fold(v, (int)nb, op);
    v = skl_shfl(v, 0);
    a2 = h2 ? op(a2, v) : v;
    h2 = true;
  }
  __syncthreads();  // s_w / s_h reused
  if (lane == 0) {
    s_h[warp] = h2;
    if (h2) s_w[warp] = a2;
  }
  __syncthreads();
  if (threadIdx.x == 0) {
    SKL_T r = s_w[0];
    for (int i = 1; i < SKL_NW; ++i)
      if (s_h[i]) r = op(r, s_w[i]);
    *result = r;
    *counter = 0u;  // ready for the next launch (stream-ordered)
  }
}

extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_reduce_vec(const SKL_T* __restrict__ in, skl_u64 n, skl_u64 wseg, SKL_T* partials,
               unsigned* counter, SKL_T* result) {
  skl_reduce_body<SKL_RVEC>(SklLoadPlain{in}, n, wseg, partials, counter, result);
}
extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_reduce_sc(const SKL_T* __restrict__ in, skl_u64 n, skl_u64 wseg, SKL_T* partials,
              unsigned* counter, SKL_T* result) {
  skl_reduce_body<1>(SklLoadPlain{in}, n, wseg, partials, counter, result);
}

#if SKL_FUSED
extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_reduce_zip_vec(const SKL_ZL* __restrict__ l, const SKL_ZR* __restrict__ r, skl_u64 n, skl_u64 wseg,
                   SKL_T* partials, unsigned* counter, SKL_T* result) {
  skl_reduce_body<SKL_RVEC>(SklLoadZip{l, r}, n, wseg, partials, counter, result);
}
extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_reduce_zip_sc(const SKL_ZL* __restrict__ l, const SKL_ZR* __restrict__ r, skl_u64 n, skl_u64 wseg,
                  SKL_T* partials, unsigned* counter, SKL_T* result) {
  skl_reduce_body<1>(SklLoadZip{l, r}, n, wseg, partials, counter, result);
}
#endif

// Ordered fold of `nrep` staged values per element (copy(+) -> block combine,
// reading A25; and the cross-GPU fold of Reduce partials): out[i] =
// s[0][i] (+) s[1][i] (+) ... (+) s[nrep-1][i], GPU order.
// All replicas' loads of an element (up to SKL_CMAXR) are issued before the
// fold, so a thread has nrep loads in flight instead of one round trip per
// replica; with `vec` (stride a multiple of SKL_RVEC, 16-byte aligned buffers)
// every load and store is 16 bytes wide.
#define SKL_CMAXR 8
template <int V>
__device__ __forceinline__ void skl_combine_run(const SKL_T* __restrict__ staging, skl_u64 stride, int nrep,
                                                SKL_T* __restrict__ out, skl_u64 n_chunks) {
  SklOp op;
  for (skl_u64 i = (skl_u64)blockIdx.x * SKL_BLOCK + threadIdx.x; i < n_chunks;
       i += (skl_u64)gridDim.x * SKL_BLOCK) {
    SklChunk<SKL_T, V> x[SKL_CMAXR];
#pragma unroll
    for (int r = 0; r < SKL_CMAXR; ++r)
      if (r < nrep) {
        if (V > 1) {
          x[r].q[0] = skl_ld16(staging + (skl_u64)r * stride + i * V);
        } else {
          x[r].e[0] = staging[(skl_u64)r * stride + i];
        }
      }
    SklChunk<SKL_T, V> a = x[0];
#pragma unroll
    for (int r = 1; r < SKL_CMAXR; ++r)
      if (r < nrep) {
#pragma unroll
        for (int k = 0; k < V; ++k) a.e[k] = op(a.e[k], x[r].e[k]);
      }
    for (int r = SKL_CMAXR; r < nrep; ++r)  // more than SKL_CMAXR devices
#pragma unroll
      for (int k = 0; k < V; ++k) a.e[k] = op(a.e[k], staging[(skl_u64)r * stride + i * V + k]);
    if (V > 1) skl_st16(out + i * V, a.q[0]);
    else out[i] = a.e[0];
  }
}
extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_combine(const SKL_T* __restrict__ staging, skl_u64 stride, int nrep, SKL_T* __restrict__ out,
            skl_u64 n, int vec) {
#if SKL_RVEC > 1
  if (vec) {
    const skl_u64 nc = n / SKL_RVEC;
    skl_combine_run<SKL_RVEC>(staging, stride, nrep, out, nc);
    // scalar tail (< SKL_RVEC elements), block 0
    const skl_u64 t0 = nc * SKL_RVEC;
    if (blockIdx.x == 0 && threadIdx.x < n - t0) {
      SklOp op;
      const skl_u64 i = t0 + threadIdx.x;
      SKL_T a = staging[i];
      for (int r = 1; r < nrep; ++r) a = op(a, staging[(skl_u64)r * stride + i]);
      out[i] = a;
    }
    return;
  }
#endif
  (void)vec;
  skl_combine_run<1>(staging, stride, nrep, out, n);
}

// copy(+) -> block fused with its exchange (reading A25; one process driving
// every device): device g folds its block slice straight out of every replica
// (peer loads over NVLink, or the same GPU for logical devices) in device order,
// out[i] = src[0][i] (+) src[1][i] (+) ... (+) src[nrep-1][i], and writes the
// result in place into its own replica - a reduce-scatter with the user's
// operator in one kernel, no staging copy.  In place is safe: device g writes
// only its own slice of its own replica, which no other device reads.
//
// One pass, no grid-stride loop: thread t of block b owns the SKL_CUNR 16-byte
// chunks b * SKL_CBLOCK * SKL_CUNR + u * SKL_CBLOCK + t (u < SKL_CUNR), issues
// every replica's loads of all of them before the first fold (in groups of 4
// replicas to bound registers) and stores the folded chunks.  Chunk indices are
// 32-bit (the host checks the count).  The previous grid-stride loop with 64-bit
// indices and a 64-bit float conversion per chunk executed ~350 instructions
// per 16-byte chunk (ncu): issue-bound at 2.7 TB/s.
#ifndef SKL_CBLOCK
#error "SKL_CBLOCK (kCombineBlock, skl_internal.h) must be defined by the program source"
#endif
#ifndef SKL_CUNR
#define SKL_CUNR 2
#endif
struct SklSrcs {
  const SKL_T* p[SKL_CMAXR];
};
// fold the SKL_CUNR chunks of this thread over every replica into a[]
template <int V>
__device__ __forceinline__ void skl_combine_fold(const SklSrcs& s, int nrep, unsigned i0, unsigned n_chunks,
                                                 SklChunk<SKL_T, V> (&a)[SKL_CUNR]) {
  SklOp op;
#pragma unroll
  for (int g0 = 0; g0 < SKL_CMAXR; g0 += 4) {
    if (g0 >= nrep) break;
    SklChunk<SKL_T, V> x[SKL_CUNR][4];
#pragma unroll
    for (int u = 0; u < SKL_CUNR; ++u) {
      const unsigned i = i0 + (unsigned)u * SKL_CBLOCK;
      if (i < n_chunks) {
#pragma unroll
        for (int j = 0; j < 4; ++j)
          if (g0 + j < nrep) {
            if (V > 1) x[u][j].q[0] = skl_ld16(s.p[g0 + j] + (size_t)i * V);
            else x[u][j].e[0] = s.p[g0 + j][i];
          }
      }
    }
#pragma unroll
    for (int u = 0; u < SKL_CUNR; ++u)
#pragma unroll
      for (int j = 0; j < 4; ++j)
        if (g0 + j < nrep) {
          if (g0 + j == 0) {
            a[u] = x[u][0];
          } else {
#pragma unroll
            for (int k = 0; k < V; ++k) a[u].e[k] = op(a[u].e[k], x[u][j].e[k]);
          }
        }
  }
}
template <int V>
__device__ __forceinline__ void skl_combine_peer_run(const SklSrcs& s, int nrep, SKL_T* out, unsigned n_chunks) {
  const unsigned i0 = blockIdx.x * (unsigned)(SKL_CBLOCK * SKL_CUNR) + threadIdx.x;
  SklChunk<SKL_T, V> a[SKL_CUNR];
  skl_combine_fold<V>(s, nrep, i0, n_chunks, a);
#pragma unroll
  for (int u = 0; u < SKL_CUNR; ++u) {
    const unsigned i = i0 + (unsigned)u * SKL_CBLOCK;
    if (i >= n_chunks) break;
    if (V > 1) skl_st16(out + (size_t)i * V, a[u].q[0]);
    else out[i] = a[u].e[0];
  }
}
// scalar fold of element i over every replica (heads and tails)
__device__ __forceinline__ SKL_T skl_combine_one(const SklSrcs& s, int nrep, skl_u64 i) {
  SklOp op;
  SKL_T a = s.p[0][i];
#pragma unroll
  for (int r = 1; r < SKL_CMAXR; ++r)   // constant indices: the pointers stay in registers
    if (r < nrep) a = op(a, s.p[r][i]);
  return a;
}
// vec: every source and out share one misalignment; the first `head` elements
// (up to the next 16-byte boundary) and the tail are folded one by one
extern "C" __global__ void __launch_bounds__(SKL_CBLOCK)
skl_combine_peer(const SklSrcs s, int nrep, SKL_T* out, skl_u64 n, int vec, int head) {
#if SKL_RVEC > 1
  if (vec) {
    const skl_u64 h = (skl_u64)head < n ? (skl_u64)head : n;
    SklSrcs sv;
#pragma unroll
    for (int r = 0; r < SKL_CMAXR; ++r) sv.p[r] = s.p[r] + h;
    const unsigned nc = (unsigned)((n - h) / SKL_RVEC);
    skl_combine_peer_run<SKL_RVEC>(sv, nrep, out + h, nc);
    const skl_u64 t0 = h + (skl_u64)nc * SKL_RVEC;
    if (blockIdx.x == 0 && threadIdx.x < h) out[threadIdx.x] = skl_combine_one(s, nrep, threadIdx.x);
    if (blockIdx.x == 0 && threadIdx.x < n - t0) out[t0 + threadIdx.x] = skl_combine_one(s, nrep, t0 + threadIdx.x);
    return;
  }
#endif
  (void)vec;
  (void)head;
  skl_combine_peer_run<1>(s, nrep, out, (unsigned)n);
}

// The same fold for logical devices sharing one GPU, in ONE launch: bases[h] is
// replica h at unit 0 (every replica covers all n elements); element e belongs
// to device e / chunk, whose replica receives the fold (chunk = the block
// distribution's ceil(units / G) units in elements; a multiple of SKL_RVEC for
// the 16-byte path).
// Replica of the device owning element e: e / chunk through a float reciprocal
// (within one of the true quotient for e < 2^31), fixed by two exact 32-bit
// compares, then selected with constant indices (the pointer table stays in
// registers).
__device__ __forceinline__ SKL_T* skl_combine_owner(const SklSrcs& s, int nrep, unsigned e, unsigned chunk,
                                                    float inv) {
  int o = (int)((float)e * inv);
  if ((unsigned)o * chunk > e) --o;
  if ((unsigned)(o + 1) * chunk <= e) ++o;
  o = o < 0 ? 0 : (o > nrep - 1 ? nrep - 1 : o);
  SKL_T* out = const_cast<SKL_T*>(s.p[0]);
#pragma unroll
  for (int r = 1; r < SKL_CMAXR; ++r)
    if (r == o) out = const_cast<SKL_T*>(s.p[r]);
  return out;
}
template <int V>
__device__ __forceinline__ void skl_combine_all_run(const SklSrcs& s, int nrep, unsigned n_chunks, unsigned chunk) {
  const unsigned i0 = blockIdx.x * (unsigned)(SKL_CBLOCK * SKL_CUNR) + threadIdx.x;
  const float inv = 1.0f / (float)chunk;
  SklChunk<SKL_T, V> a[SKL_CUNR];
  skl_combine_fold<V>(s, nrep, i0, n_chunks, a);
#pragma unroll
  for (int u = 0; u < SKL_CUNR; ++u) {
    const unsigned i = i0 + (unsigned)u * SKL_CBLOCK;
    if (i >= n_chunks) break;
    // owners of the chunk's first and last element (chunk = the block
    // distribution's unit count in elements; it need not be a multiple of V)
    const unsigned e0 = i * V;
    SKL_T* o0 = skl_combine_owner(s, nrep, e0, chunk, inv);
    if (V == 1) {
      o0[e0] = a[u].e[0];
      continue;
    }
    SKL_T* o1 = skl_combine_owner(s, nrep, e0 + V - 1, chunk, inv);
    if (o0 == o1) {
      skl_st16(o0 + e0, a[u].q[0]);
    } else {  // the chunk straddles two devices' slices
#pragma unroll
      for (int k = 0; k < V; ++k) skl_combine_owner(s, nrep, e0 + k, chunk, inv)[e0 + k] = a[u].e[k];
    }
  }
}
extern "C" __global__ void __launch_bounds__(SKL_CBLOCK)
skl_combine_all(const SklSrcs s, int nrep, skl_u64 n, skl_u64 chunk, int vec) {
#if SKL_RVEC > 1
  if (vec) {
    const unsigned nc = (unsigned)(n / SKL_RVEC);
    skl_combine_all_run<SKL_RVEC>(s, nrep, nc, (unsigned)chunk);
    const skl_u64 t0 = (skl_u64)nc * SKL_RVEC;
    if (blockIdx.x == 0 && threadIdx.x < n - t0) {
      const skl_u64 i = t0 + threadIdx.x;
      skl_combine_owner(s, nrep, (unsigned)i, (unsigned)chunk, 1.0f / (float)chunk)[i] = skl_combine_one(s, nrep, i);
    }
    return;
  }
#endif
  (void)vec;
  skl_combine_all_run<1>(s, nrep, (unsigned)n, (unsigned)chunk);
}
