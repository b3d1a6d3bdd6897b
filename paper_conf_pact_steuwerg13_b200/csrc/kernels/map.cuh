// map.cuh — Map and Zip skeleton kernels.
//
//   map f [c1..cn]          = [f(c1) .. f(cn)]
//   zip (+) [cl1..][cr1..]  = [cl1 (+) cr1 .. cln (+) crn]
//
// Configuration (#defines written by the host, skeletons.cpp):
//   SKL_TIN, SKL_TIN2 (zip), SKL_TOUT, SKL_OUT_VOID, SKL_FUNC, SKL_VEC (elements
//   per 16-byte-multiple chunk), SKL_UNROLL (chunks per thread), SKL_BLOCK,
//   SKL_XPARAMS / SKL_XARGS (extra arguments, A27).
//
// B200 design: HBM-bound, so each thread moves whole 16-byte chunks with
// ld.global.nc / st.global.cs and keeps SKL_UNROLL chunks (loads first, then
// compute, then stores) in flight; a block covers SKL_BLOCK*SKL_UNROLL
// consecutive chunks so every warp access is a contiguous 512-byte run.  The
// grid has one block per tile (hardware block scheduling balances the
// data-dependent cost of compute-bound Maps such as Mandelbrot).
#ifndef SKL_XPARAMS
#define SKL_XPARAMS
#endif
#ifndef SKL_XARGS
#define SKL_XARGS
#endif

#ifndef SKL_ILJ
#define SKL_ILJ (SKL_UNROLL * SKL_VEC)
#endif
#define SKL_QIN ((SKL_VEC * sizeof(SKL_TIN)) / 16)
#if SKL_ZIP
#define SKL_QIN2 ((SKL_VEC * sizeof(SKL_TIN2)) / 16)
#define SKL_IN2_PARAM , const SKL_TIN2* __restrict__ in2
#else
#define SKL_IN2_PARAM
#endif
#if !SKL_OUT_VOID
#define SKL_QOUT ((SKL_VEC * sizeof(SKL_TOUT)) / 16)
#define SKL_OUT_PARAM , SKL_TOUT* __restrict__ out
#else
#define SKL_OUT_PARAM , void* __restrict__ out
#endif

__device__ __forceinline__ void skl_apply_one(const SKL_TIN* __restrict__ in SKL_IN2_PARAM SKL_OUT_PARAM,
                                              skl_u64 i SKL_XPARAMS) {
#if SKL_ZIP
#if SKL_OUT_VOID
  SKL_FUNC(in[i], in2[i] SKL_XARGS);
#else
  out[i] = SKL_FUNC(in[i], in2[i] SKL_XARGS);
#endif
#else
#if SKL_OUT_VOID
  SKL_FUNC(in[i] SKL_XARGS);
#else
  out[i] = SKL_FUNC(in[i] SKL_XARGS);
#endif
#endif
}

// Vectorised kernel: requires 16-byte aligned base pointers (checked on the host).
extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_map_vec(const SKL_TIN* __restrict__ in SKL_IN2_PARAM SKL_OUT_PARAM, skl_u64 n SKL_XPARAMS) {
  const skl_u64 nch = n / SKL_VEC;
  const skl_u64 base = (skl_u64)blockIdx.x * (SKL_BLOCK * SKL_UNROLL) + threadIdx.x;
  SklChunk<SKL_TIN, SKL_VEC> a[SKL_UNROLL];
#if SKL_ZIP
  SklChunk<SKL_TIN2, SKL_VEC> b[SKL_UNROLL];
#endif
#pragma unroll
  for (int u = 0; u < SKL_UNROLL; ++u) {
    const skl_u64 c = base + (skl_u64)u * SKL_BLOCK;
    if (c < nch) {
      const char* p = (const char*)in + c * (SKL_VEC * sizeof(SKL_TIN));
#pragma unroll
      for (int q = 0; q < (int)SKL_QIN; ++q) a[u].q[q] = skl_ld16(p + 16 * q);
#if SKL_ZIP
      const char* p2 = (const char*)in2 + c * (SKL_VEC * sizeof(SKL_TIN2));
#pragma unroll
      for (int q = 0; q < (int)SKL_QIN2; ++q) b[u].q[q] = skl_ld16(p2 + 16 * q);
#endif
    }
  }
#pragma unroll
  for (int u = 0; u < SKL_UNROLL; ++u) {
    const skl_u64 c = base + (skl_u64)u * SKL_BLOCK;
    // Lanes running this chunk reconverge after every element: a customising
    // function with a data-dependent loop (LM OSEM ray walks, Mandelbrot) would
    // otherwise leave the warp split into drifting one-lane groups (independent
    // thread scheduling does not force reconvergence between unrolled calls).
    const unsigned act = __ballot_sync(SKL_FULL, c < nch);
    if (c < nch) {
#if SKL_OUT_VOID
#pragma unroll
      for (int k = 0; k < SKL_VEC; ++k) {
#if SKL_ZIP
        SKL_FUNC(a[u].e[k], b[u].e[k] SKL_XARGS);
#else
        SKL_FUNC(a[u].e[k] SKL_XARGS);
#endif
        __syncwarp(act);
      }
#else
      SklChunk<SKL_TOUT, SKL_VEC> r;
#pragma unroll
      for (int k = 0; k < SKL_VEC; ++k) {
#if SKL_ZIP
        r.e[k] = SKL_FUNC(a[u].e[k], b[u].e[k] SKL_XARGS);
#else
        r.e[k] = SKL_FUNC(a[u].e[k] SKL_XARGS);
#endif
        __syncwarp(act);
      }
      char* o = (char*)out + c * (SKL_VEC * sizeof(SKL_TOUT));
#pragma unroll
      for (int q = 0; q < (int)SKL_QOUT; ++q) skl_st16(o + 16 * q, r.q[q]);
#endif
    }
  }
  // ragged tail: the n % SKL_VEC last elements, done by the last block
  if (blockIdx.x == gridDim.x - 1) {
    const skl_u64 t = nch * SKL_VEC + threadIdx.x;
    if (threadIdx.x < SKL_VEC && t < n) {
#if SKL_ZIP
      skl_apply_one(in, in2, out, t SKL_XARGS);
#else
      skl_apply_one(in, out, t SKL_XARGS);
#endif
    }
  }
}

// Scalar kernel for unaligned views: element-wise, SKL_UNROLL per thread.
extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_map_sc(const SKL_TIN* __restrict__ in SKL_IN2_PARAM SKL_OUT_PARAM, skl_u64 n SKL_XPARAMS) {
  const skl_u64 base = (skl_u64)blockIdx.x * (SKL_BLOCK * SKL_UNROLL) + threadIdx.x;
#pragma unroll
  for (int u = 0; u < SKL_UNROLL; ++u) {
    const skl_u64 i = base + (skl_u64)u * SKL_BLOCK;
    if (i < n) {
#if SKL_ZIP
      skl_apply_one(in, in2, out, i SKL_XARGS);
#else
      skl_apply_one(in, out, i SKL_XARGS);
#endif
    }
  }
}

// Warp-interleaved kernel (skl_set_option "map_interleave" 1): for customising
// functions whose cost varies per element (Mandelbrot, ray walks).  Lane l of a
// warp handles elements base + j*32 + l, j = 0 .. SKL_UNROLL*SKL_VEC-1, so at
// every step the 32 lanes work on 32 neighbouring elements (similar cost: less
// idle-lane time than 32 lanes x SKL_VEC consecutive elements each; Mandelbrot
// 4096x3072: 6.5 % instead of 16.6 % of lane-time idle, from the oracle's
// counts).  Each load / store instruction still covers a contiguous run.
extern "C" __global__ void __launch_bounds__(SKL_BLOCK)
skl_map_il(const SKL_TIN* __restrict__ in SKL_IN2_PARAM SKL_OUT_PARAM, skl_u64 n SKL_XPARAMS) {
  constexpr int J = SKL_ILJ;  // elements per lane (option map_il_elems; default one chunk)
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const skl_u64 base = ((skl_u64)blockIdx.x * (SKL_BLOCK / 32) + warp) * (32 * J) + lane;
  SKL_TIN a[J];
#if SKL_ZIP
  SKL_TIN2 b[J];
#endif
#pragma unroll
  for (int j = 0; j < J; ++j) {
    const skl_u64 i = base + (skl_u64)j * 32;
    if (i < n) {
      a[j] = in[i];
#if SKL_ZIP
      b[j] = in2[i];
#endif
    }
  }
#pragma unroll
  for (int j = 0; j < J; ++j) {
    const skl_u64 i = base + (skl_u64)j * 32;
    const unsigned act = __ballot_sync(SKL_FULL, i < n);
    if (i < n) {
#if SKL_OUT_VOID
#if SKL_ZIP
      SKL_FUNC(a[j], b[j] SKL_XARGS);
#else
      SKL_FUNC(a[j] SKL_XARGS);
#endif
#else
#if SKL_ZIP
      out[i] = SKL_FUNC(a[j], b[j] SKL_XARGS);
#else
      out[i] = SKL_FUNC(a[j] SKL_XARGS);
#endif
#endif
      __syncwarp(act);
    }
  }
}
