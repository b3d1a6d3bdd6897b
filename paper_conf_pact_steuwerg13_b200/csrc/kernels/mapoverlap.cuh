// mapoverlap.cuh — MapOverlap skeleton, matrix and vector forms.
//
//   mout[i,j] = f( min[i-d .. i+d, j-d .. j+d] )
// f receives a pointer to the centre element and reads neighbours with
// get(p, dx, dy), dx = column offset, dy = row offset (A15).
// Out-of-bounds neighbours read a neutral value or the nearest valid element
// (A20: each coordinate clamped independently).
//
// B200 design: the paper's kernel "uses the fast local memory";
// here each block stages an output tile plus its halo in shared memory with
// coalesced 16-byte loads, resolving the boundary mode while loading (no
// per-access branch in f), then every thread applies f to a SKL_RH x SKL_CW
// register block of outputs so neighbouring calls share shared-memory reads.
// get() is a constant-offset load from the tile (SKL_PITCH is a compile-time
// row pitch).  The input part holds rows [in_row0, in_row0 + in_rows) of the
// global matrix (block rows + halo rows under the overlap distribution).
// Configuration: SKL_TIN, SKL_TOUT, SKL_FUNC, SKL_D, SKL_BOUNDARY, SKL_TH,
// SKL_TW, SKL_RH, SKL_CW, SKL_A (halo columns staged, >= d, 16-byte multiple),
// SKL_PITCH, SKL_BLOCK, SKL_MO1D.
#if SKL_DEBUG_BOUNDS
extern "C" __device__ unsigned int skl_bounds_flag = 0u;
#endif

template <int B> struct SklRaw { typedef unsigned char type; };  // unused width
template <> struct SklRaw<1> { typedef unsigned char type; };
template <> struct SklRaw<2> { typedef unsigned short type; };
template <> struct SklRaw<4> { typedef unsigned int type; };
template <> struct SklRaw<8> { typedef uint2 type; };
template <> struct SklRaw<16> { typedef uint4 type; };

#define SKL_EPC (16 / (int)sizeof(SKL_TIN))
// SKL_OUTB = SKL_CW * sizeof(SKL_TOUT), written by the host (used in #if)
#define SKL_OUT_PACK (SKL_OUTB == 1 || SKL_OUTB == 2 || SKL_OUTB == 4 || SKL_OUTB == 8 || SKL_OUTB == 16)

__device__ __forceinline__ long skl_clampl(long v, long lo, long hi) {
  return v < lo ? lo : (v > hi ? hi : v);
}

union SklMoRes {
  SKL_TOUT e[SKL_CW];
  typename SklRaw<SKL_OUTB>::type raw;
};
// four byte results -> one 32-bit word with three byte permutes (PRMT); the
// union's bytewise assembly took five shift/mask instructions per word
__device__ __forceinline__ unsigned skl_pack4(unsigned b0, unsigned b1, unsigned b2, unsigned b3) {
  return __byte_perm(__byte_perm(b0, b1, 0x3340), __byte_perm(b2, b3, 0x3340), 0x5410);
}
// store one thread's SKL_CW outputs of a row at o (ncols columns remain in the row)
__device__ __forceinline__ void skl_mo_store(SKL_TOUT* o, const SklMoRes& v, bool full, long ncols) {
#if SKL_OUT_PACK
  if (full) {
#if SKL_SO == 1 && SKL_CW % 4 == 0
    unsigned w[SKL_CW / 4];
#pragma unroll
    for (int k = 0; k < SKL_CW / 4; ++k)
      w[k] = skl_pack4((unsigned char)v.e[4 * k], (unsigned char)v.e[4 * k + 1], (unsigned char)v.e[4 * k + 2],
                       (unsigned char)v.e[4 * k + 3]);
#if SKL_CW == 16
    *(uint4*)o = make_uint4(w[0], w[1], w[2], w[3]);
#elif SKL_CW == 8
    *(uint2*)o = make_uint2(w[0], w[1]);
#else
    *(unsigned*)o = w[0];
#endif
#else
    *(typename SklRaw<SKL_OUTB>::type*)o = v.raw;
#endif
    return;
  }
#endif
#pragma unroll
  for (int j = 0; j < SKL_CW; ++j)
    if (j < ncols) o[j] = v.e[j];
}

#if !SKL_MO1D
// ------------------------------------------------------------------ 2-D
#define SKL_SROWS (SKL_TH + 2 * SKL_D)
#define SKL_CPR (SKL_PITCH / SKL_EPC)  // 16-byte chunks per smem row

#ifndef SKL_MO_MINB
#define SKL_MO_MINB 1
#endif
#ifndef SKL_MO_HEAVY
#define SKL_MO_HEAVY 0
#endif

// Geometry of one launch: 32-bit row / column arithmetic (the host guarantees
// R, C < 2^31); 64-bit only where a row index is scaled to an element offset.
struct SklMoGeo {
  int Ri, Ci, rb, re, irow0, orow0, hd;
};

// Stage the input window of the tile at (r0, c0) into `tile`: rows r0-d ..
// r0+TH+d-1, columns c0-A .. c0+TW+A-1.  Issues cp.async copies (the caller
// commits / waits) and plain stores for border chunks.
__device__ __forceinline__ void skl_mo_stage(SKL_TIN* tile, const SKL_TIN* __restrict__ in, const SklMoGeo& G,
                                             int r0, int c0, SKL_TIN neutral, int vec_ok) {
  const int Ri = G.Ri, Ci = G.Ci;
  const bool interior = vec_ok && c0 - SKL_A >= 0 && c0 + SKL_TW + SKL_A <= Ci && r0 - SKL_D >= 0 &&
                        r0 + SKL_TH + SKL_D <= Ri && r0 + SKL_TH <= G.re;
  if (interior) {
    // block-uniform fast path: every staged chunk is an in-range 16-byte copy.
    // The tile is dense in shared memory (SKL_PITCH = SKL_CPR chunks), so chunk
    // q lands at byte 16 q; its global address advances by a constant per step
    // (plus one row's remainder when the column wraps)
    const int jc0 = threadIdx.x % SKL_CPR;
    const char* gp = (const char*)(in + (long)(r0 - SKL_D - G.irow0 + (int)threadIdx.x / SKL_CPR) * Ci +
                                   (c0 - SKL_A) + jc0 * SKL_EPC);
    unsigned sa = (unsigned)__cvta_generic_to_shared(tile) + 16u * threadIdx.x;
    const long rowb = (long)Ci * (long)sizeof(SKL_TIN);
    const long step = (long)(SKL_BLOCK / SKL_CPR) * rowb + (long)(SKL_BLOCK % SKL_CPR) * 16;
    const long wrap = rowb - (long)SKL_CPR * 16;
    int jc = jc0;
#pragma unroll 4
    for (int q = threadIdx.x; q < SKL_SROWS * SKL_CPR; q += SKL_BLOCK) {
      asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" ::"r"(sa), "l"(gp) : "memory");
      sa += 16u * SKL_BLOCK;
      gp += step;
      jc += SKL_BLOCK % SKL_CPR;
      if (jc >= SKL_CPR) {
        jc -= SKL_CPR;
        gp += wrap;
      }
    }
    return;
  }
  for (int q = threadIdx.x; q < SKL_SROWS * SKL_CPR; q += SKL_BLOCK) {
    const int i = q / SKL_CPR, jc = q - i * SKL_CPR;
    int gr = r0 - SKL_D + i;
    const int gc0 = c0 - SKL_A + jc * SKL_EPC;
    const bool row_in = gr >= 0 && gr < Ri;
#if SKL_BOUNDARY == 1
    gr = gr < 0 ? 0 : (gr > Ri - 1 ? Ri - 1 : gr);
#endif
    SKL_TIN* dst = tile + i * SKL_PITCH + jc * SKL_EPC;
    if (r0 - SKL_D + i >= G.re + SKL_D) {  // below the last output row's window: unused
#pragma unroll
      for (int e = 0; e < SKL_EPC; ++e) dst[e] = neutral;
      continue;
    }
    const SKL_TIN* row = in + (long)(gr - G.irow0) * Ci;
    if (vec_ok && (SKL_BOUNDARY == 1 || row_in) && gc0 >= 0 && gc0 + SKL_EPC <= Ci) {
      // asynchronous 16-byte global->shared copy (LDGSTS), no register round trip
      const unsigned sa = (unsigned)__cvta_generic_to_shared(dst);
      asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" ::"r"(sa), "l"(row + gc0) : "memory");
    } else {
#pragma unroll
      for (int e = 0; e < SKL_EPC; ++e) {
        int gc = gc0 + e;
        SKL_TIN v;
#if SKL_BOUNDARY == 1
        gc = gc < 0 ? 0 : (gc > Ci - 1 ? Ci - 1 : gc);
        v = row[gc];
#else
        if (row_in && gc >= 0 && gc < Ci) v = row[gc];
        else v = neutral;
#endif
        dst[e] = v;
      }
    }
  }
}

// Apply f to the staged tile: a SKL_RH x SKL_CW block of outputs per thread.
__device__ __forceinline__ void skl_mo_apply(const SKL_TIN* tile, SKL_TOUT* __restrict__ out, const SklMoGeo& G,
                                             int r0, int c0, int vec_ok, SKL_TOUT* __restrict__ push_up,
                                             SKL_TOUT* __restrict__ push_down) {
  const int Ci = G.Ci, rb = G.rb, re = G.re, hdi = G.hd;
  const int ty = threadIdx.x / (SKL_TW / SKL_CW), tx = threadIdx.x % (SKL_TW / SKL_CW);
  const int cc = c0 + tx * SKL_CW;
  const int ncols = Ci - cc;                        // columns left in the row from cc
  const bool full = vec_ok && ncols >= SKL_CW;      // whole packed store in range
  const int rt = r0 + ty * SKL_RH;                  // this thread's first row
  SKL_TOUT* o = out + (long)(rt - G.orow0) * Ci + cc;
  // fused halo push: the first / last hd rows of this device's
  // block also go into the neighbours' halo rows (peer memory), so the next
  // overlap read needs no exchange.  Block-uniform; the common path below
  // carries none of it (live registers matter: f may call the IEEE sqrt
  // subroutine).
  if ((push_up && r0 < rb + hdi) || (push_down && r0 + SKL_TH > re - hdi)) {
#pragma unroll
    for (int i = 0; i < SKL_RH; ++i) {
      const int r = rt + i;
      const SKL_TIN* p = tile + (SKL_D + ty * SKL_RH + i) * SKL_PITCH + SKL_A + tx * SKL_CW;
      SklMoRes res;
#pragma unroll
      for (int j = 0; j < SKL_CW; ++j) res.e[j] = SKL_FUNC((SKL_TIN*)(p + j));
      if (r >= re) continue;
      skl_mo_store(o + (long)i * Ci, res, full, ncols);
      if (push_up && r < rb + hdi) skl_mo_store(push_up + (long)(r - rb) * Ci + cc, res, full, ncols);
      if (push_down && r >= re - hdi)
        skl_mo_store(push_down + (long)(r - (re - hdi)) * Ci + cc, res, full, ncols);
    }
    return;
  }
#if SKL_OUT_PACK && SKL_MO_HEAVY
  if (full && rt + SKL_RH <= re) {
    // every row of this thread in range and whole packed stores (all threads
    // but those of a device's last tile row or the matrix's last columns): no
    // per-row guard or partial-store path in the loop.  Heavy functions only
    // (the Gaussian 117 -> 109 us, Listing 1.5's Sobel 76 -> 74 us); for a
    // light one the second copy of the loop cost more than the guards
    // (identity u8 26.7 -> 27.7 us)
#pragma unroll
    for (int i = 0; i < SKL_RH; ++i) {
      const SKL_TIN* p = tile + (SKL_D + ty * SKL_RH + i) * SKL_PITCH + SKL_A + tx * SKL_CW;
      SklMoRes res;
#pragma unroll
      for (int j = 0; j < SKL_CW; ++j) res.e[j] = SKL_FUNC((SKL_TIN*)(p + j));
      skl_mo_store(o + (long)i * Ci, res, true, SKL_CW);
    }
    return;
  }
#endif
#pragma unroll
  for (int i = 0; i < SKL_RH; ++i) {
    const SKL_TIN* p = tile + (SKL_D + ty * SKL_RH + i) * SKL_PITCH + SKL_A + tx * SKL_CW;
    SklMoRes res;
#pragma unroll
    // f may declare a non-const pointer (Listing 1.2: "float func(float* m_in)")
    for (int j = 0; j < SKL_CW; ++j) res.e[j] = SKL_FUNC((SKL_TIN*)(p + j));
    if (rt + i < re) skl_mo_store(o + (long)i * Ci, res, full, ncols);
  }
}

// One block per tile (grid = tiles_x x tiles_y).
extern "C" __global__ void __launch_bounds__(SKL_BLOCK, SKL_MO_MINB)
skl_mo2d(const SKL_TIN* __restrict__ in, long in_row0, long in_rows, SKL_TOUT* __restrict__ out,
         long out_row0, long R, long C, long r_begin, long r_end, SKL_TIN neutral, int vec_ok,
         SKL_TOUT* __restrict__ push_up, SKL_TOUT* __restrict__ push_down, long hd) {
  __shared__ __align__(16) SKL_TIN tile[SKL_SROWS * SKL_PITCH];
  const SklMoGeo G{(int)R, (int)C, (int)r_begin, (int)r_end, (int)in_row0, (int)out_row0, (int)hd};
  const int r0 = G.rb + (int)blockIdx.y * SKL_TH;
  const int c0 = (int)blockIdx.x * SKL_TW;
  skl_mo_stage(tile, in, G, r0, c0, neutral, vec_ok);
  asm volatile("cp.async.wait_all;" ::: "memory");
  __syncthreads();
  skl_mo_apply(tile, out, G, r0, c0, vec_ok, push_up, push_down);
  (void)in_rows;
}

// TMA staging (option mo_tma, the default where a tensor map can describe the
// part): one thread stages the block's whole (TH + 2d) x PITCH window with a
// single cp.async.bulk.tensor.2d (out-of-matrix cells zero-filled by the copy
// engine, NEAREST / non-zero neutral border tiles patched in shared memory),
// the block waits on an mbarrier and applies f as skl_mo2d does.  The per-thread
// staging walk (address arithmetic and one cp.async per 16 bytes, plus the
// general path for border tiles) was ~40 % of the instructions of a byte stencil
// (ncu of the identity u8 stencil: 258 instructions per warp for 32 outputs
// per thread).  x coordinates are in 2^ushift-byte units.
struct alignas(64) SklTmap {
  unsigned long long opaque[16];
};
__device__ __forceinline__ void skl_mbar_wait(unsigned a, unsigned parity) {
  unsigned done;
  do {
    asm volatile(
        "{ .reg .pred p; mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2; selp.u32 %0, 1, 0, p; }"
        : "=r"(done) : "r"(a), "r"(parity) : "memory");
  } while (!done);
}
// Out-of-matrix cells of a TMA-staged tile (zero-filled) get the boundary mode's
// value: NEAREST copies the nearest in-matrix row, then column (each coordinate
// clamped independently, A20); NEUTRAL writes the neutral value.  All nthr
// threads of the block (named barrier 1) take part.
template <int NT>
__device__ __forceinline__ void skl_mo_fix(SKL_TIN* tile, const SklMoGeo& G, int r0, int c0, SKL_TIN neutral) {
  const int gr0 = r0 - SKL_D, gc0 = c0 - SKL_A;
  const int top = gr0 < 0 ? -gr0 : 0, bot = G.Ri - gr0;  // rows [top, bot) are inside
  const int left = gc0 < 0 ? -gc0 : 0, right = G.Ci - gc0;
#if SKL_BOUNDARY == 1
  if (top > 0 || bot < SKL_SROWS) {
    for (int q = threadIdx.x; q < SKL_SROWS * SKL_PITCH; q += NT) {
      const int i = q / SKL_PITCH, j = q - i * SKL_PITCH;
      if (i < top) tile[q] = tile[top * SKL_PITCH + j];
      else if (i >= bot) tile[q] = tile[(bot - 1) * SKL_PITCH + j];
    }
    asm volatile("bar.sync 1, %0;" ::"n"(NT) : "memory");
  }
  if (left > 0 || right < SKL_PITCH) {
    for (int q = threadIdx.x; q < SKL_SROWS * SKL_PITCH; q += NT) {
      const int i = q / SKL_PITCH, j = q - i * SKL_PITCH;
      if (j < left) tile[q] = tile[i * SKL_PITCH + left];
      else if (j >= right) tile[q] = tile[i * SKL_PITCH + right - 1];
    }
  }
#else
  for (int q = threadIdx.x; q < SKL_SROWS * SKL_PITCH; q += NT) {
    const int i = q / SKL_PITCH, j = q - i * SKL_PITCH;
    if (i < top || i >= bot || j < left || j >= right) tile[q] = neutral;
  }
#endif
  asm volatile("bar.sync 1, %0;" ::"n"(NT) : "memory");
}

// SKL_MO_KT tiles per block, stacked vertically (compile-time; option mo_kt):
// thread 0 issues all their TMA copies at once, so the later tiles arrive while
// f runs on the first (the tile wait was 29 % of the Gaussian's stall samples
// with one tile per block); every tile has its own buffer and mbarrier.  (A
// run-time tile count around the inlined f made ptxas spill the byte stencils
// heavily - 4x slower - so the count is a compile-time constant.)
#ifndef SKL_MO_KT
#define SKL_MO_KT 1
#endif
extern "C" __global__ void __launch_bounds__(SKL_BLOCK, SKL_MO_MINB)
skl_mo2d_t(const __grid_constant__ SklTmap tmap, SKL_TOUT* __restrict__ out, long in_row0, long out_row0, long R,
           long C, long r_begin, long r_end, SKL_TIN neutral, int vec_ok, SKL_TOUT* __restrict__ push_up,
           SKL_TOUT* __restrict__ push_down, long hd, int fix, int ushift) {
  constexpr unsigned TB = SKL_SROWS * SKL_PITCH * (unsigned)sizeof(SKL_TIN);
  constexpr unsigned TS = (TB + 127u) / 128u * 128u;
#if SKL_MO_KT == 1
  __shared__ __align__(128) SKL_TIN skl_tile0[SKL_SROWS * SKL_PITCH];
  unsigned char* smem = (unsigned char*)skl_tile0;
#else
  extern __shared__ __align__(128) unsigned char skl_mo_dyn[];  // SKL_MO_KT x TS (+128 to align)
  unsigned char* smem = skl_mo_dyn + ((128u - ((unsigned)__cvta_generic_to_shared(skl_mo_dyn) & 127u)) & 127u);
#endif
  __shared__ __align__(8) unsigned long long bars[SKL_MO_KT];
  const SklMoGeo G{(int)R, (int)C, (int)r_begin, (int)r_end, (int)in_row0, (int)out_row0, (int)hd};
  const int rt0 = G.rb + (int)blockIdx.y * (SKL_TH * SKL_MO_KT);
  const int c0 = (int)blockIdx.x * SKL_TW;
  const unsigned b0 = (unsigned)__cvta_generic_to_shared(bars);
  const unsigned sbase = (unsigned)__cvta_generic_to_shared(smem);
  if (threadIdx.x == 0) {
#pragma unroll
    for (int k = 0; k < SKL_MO_KT; ++k)
      asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(b0 + 8u * k) : "memory");
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
#pragma unroll
    for (int k = 0; k < SKL_MO_KT; ++k) {
      const int r0 = rt0 + k * SKL_TH;
      if (r0 >= G.re) break;
      asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(b0 + 8u * k), "n"(TB) : "memory");
      asm volatile(
          "cp.async.bulk.tensor.2d.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3}], "
          "[%4];" ::"r"(sbase + TS * k),
          "l"((unsigned long long)&tmap), "r"(((c0 - SKL_A) * (int)sizeof(SKL_TIN)) >> ushift),
          "r"(r0 - SKL_D - G.irow0), "r"(b0 + 8u * k)
          : "memory");
    }
  }
  __syncthreads();  // the barriers are initialised before anyone waits on them
#pragma unroll 1
  for (int k = 0; k < SKL_MO_KT; ++k) {
    const int r0 = rt0 + k * SKL_TH;
    if (r0 >= G.re) break;
    SKL_TIN* tile = (SKL_TIN*)(smem + TS * k);
    skl_mbar_wait(b0 + 8u * k, 0);
    if (fix && (r0 - SKL_D < 0 || r0 + SKL_TH + SKL_D > G.Ri || c0 - SKL_A < 0 || c0 + SKL_TW + SKL_A > G.Ci))
      skl_mo_fix<SKL_BLOCK>(tile, G, r0, c0, neutral);
    skl_mo_apply(tile, out, G, r0, c0, vec_ok, push_up, push_down);
  }
}

// Persistent variant: a grid of resident blocks walks the tiles (t = blockIdx.x,
// + gridDim.x, ...) with two shared-memory buffers, staging tile k+1 while
// applying f to tile k, so the load latency of a tile hides behind the
// computation of the previous one (ncu of the one-tile-per-block kernel: the
// top stall was the wait for the tile, with only 4 blocks resident per SM).
extern "C" __global__ void __launch_bounds__(SKL_BLOCK, SKL_MO_MINB)
skl_mo2d_p(const SKL_TIN* __restrict__ in, long in_row0, long in_rows, SKL_TOUT* __restrict__ out,
           long out_row0, long R, long C, long r_begin, long r_end, SKL_TIN neutral, int vec_ok,
           SKL_TOUT* __restrict__ push_up, SKL_TOUT* __restrict__ push_down, long hd, int tiles_x, int ntiles) {
  extern __shared__ __align__(16) unsigned char skl_mo_dyn[];
  SKL_TIN* buf[2] = {(SKL_TIN*)skl_mo_dyn, (SKL_TIN*)skl_mo_dyn + SKL_SROWS * SKL_PITCH};
  const SklMoGeo G{(int)R, (int)C, (int)r_begin, (int)r_end, (int)in_row0, (int)out_row0, (int)hd};
  int t = blockIdx.x;
  if (t >= ntiles) return;
  skl_mo_stage(buf[0], in, G, G.rb + (t / tiles_x) * SKL_TH, (t % tiles_x) * SKL_TW, neutral, vec_ok);
  asm volatile("cp.async.commit_group;" ::: "memory");
  for (int k = 0; t < ntiles; ++k, t += gridDim.x) {
    const int tn = t + gridDim.x;
    if (tn < ntiles)
      skl_mo_stage(buf[(k + 1) & 1], in, G, G.rb + (tn / tiles_x) * SKL_TH, (tn % tiles_x) * SKL_TW, neutral,
                   vec_ok);
    asm volatile("cp.async.commit_group;" ::: "memory");
    asm volatile("cp.async.wait_group 1;" ::: "memory");  // tile t has landed
    __syncthreads();
    skl_mo_apply(buf[k & 1], out, G, G.rb + (t / tiles_x) * SKL_TH, (t % tiles_x) * SKL_TW, vec_ok, push_up,
                 push_down);
    __syncthreads();  // buf[k & 1] is restaged two tiles later
  }
  (void)in_rows;
}

// ------------------------------------------------------------------ 2-D, TMA + warp specialisation
// Persistent resident blocks of SKL_BLOCK consumer threads plus one producer
// warp.  The producer's elected lane stages tile after tile with one TMA box
// copy each (cp.async.bulk.tensor.2d: the whole (TH + 2d) x PITCH window in one
// instruction, out-of-matrix cells zero-filled by the copy engine) into a ring
// of nstages shared-memory buffers, signalling a "full" mbarrier by transaction
// bytes; the consumers wait on it, apply f exactly as skl_mo2d does
// (skl_mo_apply) and release the buffer through an "empty" mbarrier (one arrival
// per consumer warp).  Consumer threads issue no staging instructions and the
// next tiles' loads are always in flight while f runs.  Border tiles whose
// boundary mode is not "zero" (NEAREST, or NEUTRAL with a non-zero value) are
// patched in shared memory by the consumers before f runs.
#define SKL_WS_MAXS 8
#ifndef SKL_WS_MINB
#define SKL_WS_MINB 1
#endif
__device__ __forceinline__ void skl_bar_consumers() {
  asm volatile("bar.sync 1, %0;" ::"n"(SKL_BLOCK) : "memory");
}

extern "C" __global__ void __launch_bounds__(SKL_BLOCK + 32, SKL_WS_MINB)
skl_mo2d_ws(const __grid_constant__ SklTmap tmap, SKL_TOUT* __restrict__ out, long in_row0, long out_row0,
            long R, long C, long r_begin, long r_end, SKL_TIN neutral, int vec_ok, SKL_TOUT* __restrict__ push_up,
            SKL_TOUT* __restrict__ push_down, long hd, int tiles_x, int ntiles, int nstages, int fix, int ushift) {
  extern __shared__ __align__(128) unsigned char skl_mo_dyn[];
  __shared__ __align__(8) unsigned long long bars[2 * SKL_WS_MAXS];
  constexpr unsigned TB = SKL_SROWS * SKL_PITCH * (unsigned)sizeof(SKL_TIN);
  constexpr unsigned TS = (TB + 127u) / 128u * 128u;  // TMA destinations are 128-byte aligned
  const SklMoGeo G{(int)R, (int)C, (int)r_begin, (int)r_end, (int)in_row0, (int)out_row0, (int)hd};
  const unsigned raw = (unsigned)__cvta_generic_to_shared(skl_mo_dyn);
  const unsigned base = (raw + 127u) & ~127u;
  const unsigned full0 = (unsigned)__cvta_generic_to_shared(bars), empty0 = full0 + 8u * SKL_WS_MAXS;
  if (threadIdx.x == 0) {
    for (int s = 0; s < nstages; ++s) {
      asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(full0 + 8u * s) : "memory");
      asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(empty0 + 8u * s), "n"(SKL_BLOCK / 32)
                   : "memory");
    }
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  if (warp == SKL_BLOCK / 32) {  // producer
    if (lane == 0) {
      int k = 0;
      for (int t = blockIdx.x; t < ntiles; t += gridDim.x, ++k) {
        const int s = k % nstages;
        if (k >= nstages) skl_mbar_wait(empty0 + 8u * s, ((k / nstages) & 1) ^ 1);
        asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(full0 + 8u * s), "n"(TB)
                     : "memory");
        const int r0 = G.rb + (t / tiles_x) * SKL_TH, c0 = (t % tiles_x) * SKL_TW;
        asm volatile(
            "cp.async.bulk.tensor.2d.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3}], "
            "[%4];" ::"r"(base + TS * s),
            "l"((unsigned long long)&tmap), "r"(((c0 - SKL_A) * (int)sizeof(SKL_TIN)) >> ushift), "r"(r0 - SKL_D - G.irow0),
            "r"(full0 + 8u * s)
            : "memory");
      }
    }
    return;
  }
  int k = 0;
  for (int t = blockIdx.x; t < ntiles; t += gridDim.x, ++k) {
    const int s = k % nstages;
    skl_mbar_wait(full0 + 8u * s, (k / nstages) & 1);
    SKL_TIN* tile = (SKL_TIN*)(skl_mo_dyn + (base - raw) + TS * s);
    const int r0 = G.rb + (t / tiles_x) * SKL_TH, c0 = (t % tiles_x) * SKL_TW;
    const bool border = fix && (r0 - SKL_D < 0 || r0 + SKL_TH + SKL_D > G.Ri || c0 - SKL_A < 0 ||
                                c0 + SKL_TW + SKL_A > G.Ci);
    if (border) skl_mo_fix<SKL_BLOCK>(tile, G, r0, c0, neutral);
    skl_mo_apply(tile, out, G, r0, c0, vec_ok, push_up, push_down);
    // generic-proxy writes of the patch must be ordered before the next TMA write
    if (border) asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
    __syncwarp();
    if (lane == 0) asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(empty0 + 8u * s) : "memory");
  }
}
#else
// ------------------------------------------------------------------ 1-D (vector)
#define SKL_SLEN (SKL_TW + 2 * SKL_A)
extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_mo1d(const SKL_TIN* __restrict__ in, long in_lo, long in_n, SKL_TOUT* __restrict__ out,
         long out_lo, long N, long unused, long i_begin, long i_end, SKL_TIN neutral, int vec_ok,
         SKL_TOUT* __restrict__ push_up, SKL_TOUT* __restrict__ push_down, long hd) {
  __shared__ __align__(16) SKL_TIN tile[SKL_SLEN];
  const long e0 = i_begin + (long)blockIdx.x * SKL_TW;
  for (int q = threadIdx.x; q < SKL_SLEN / SKL_EPC; q += SKL_BLOCK) {
    const long g0 = e0 - SKL_A + (long)q * SKL_EPC;
    SKL_TIN* dst = tile + q * SKL_EPC;
    if (vec_ok && g0 >= in_lo && g0 + SKL_EPC <= in_lo + in_n && g0 >= 0 && g0 + SKL_EPC <= N &&
        ((g0 - in_lo) % SKL_EPC) == 0) {
      const unsigned sa = (unsigned)__cvta_generic_to_shared(dst);
      asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" ::"r"(sa), "l"(in + (g0 - in_lo)) : "memory");
    } else {
#pragma unroll
      for (int e = 0; e < SKL_EPC; ++e) {
        long g = g0 + e;
        SKL_TIN v;
#if SKL_BOUNDARY == 1
        g = skl_clampl(g, 0, N - 1);
        if (g >= in_lo && g < in_lo + in_n) v = in[g - in_lo];
        else v = neutral;  // outside every needed window
#else
        if (g >= 0 && g < N && g >= in_lo && g < in_lo + in_n) v = in[g - in_lo];
        else v = neutral;
#endif
        dst[e] = v;
      }
    }
  }
  asm volatile("cp.async.wait_all;" ::: "memory");
  __syncthreads();
  const long i0 = e0 + (long)threadIdx.x * SKL_CW;
  const SKL_TIN* p = tile + SKL_A + threadIdx.x * SKL_CW;
#pragma unroll
  for (int j = 0; j < SKL_CW; ++j) {
    const long i = i0 + j;
    if (i < i_end) {
      const SKL_TOUT v = SKL_FUNC((SKL_TIN*)(p + j));
      out[i - out_lo] = v;
      if (push_up && i < i_begin + hd) push_up[i - i_begin] = v;          // fused halo push
      if (push_down && i >= i_end - hd) push_down[i - (i_end - hd)] = v;
    }
  }
  (void)unused;
}
#endif
