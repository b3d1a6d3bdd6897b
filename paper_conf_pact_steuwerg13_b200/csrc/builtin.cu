// builtin.cu — the kernels that need no customising function: filling a
// container's device parts with a value (skl_fill; used to zero the copy(+)
// image replicas of LM OSEM before every subset, reading A25), and the batched
// transfer kernel that executes all moves of a redistribution into one device
// in a single launch (halo refresh P:L214-222).  Compiled by nvcc
// for sm_100a into libskl.so.
#include "skl_internal.h"

namespace skl {

struct FillPattern {
  unsigned char b[64];
};

// 16-byte stores of a 16-byte pattern (element size divides 16), byte tail.
// The tail bytes come from the pattern word itself (it repeats every 16 bytes):
// indexing the by-value pattern array would copy it to local memory in every
// thread (64 B of stack traffic per thread, measured 4x slower).
__device__ __forceinline__ unsigned char skl_pat_byte(const uint4& v, unsigned i) {
  const unsigned w = (i & 15u) >> 2;
  const unsigned x = w == 0 ? v.x : (w == 1 ? v.y : (w == 2 ? v.z : v.w));
  return (unsigned char)(x >> (8u * (i & 3u)));
}
__global__ void __launch_bounds__(256) skl_fill16(uint4* __restrict__ dst, size_t n16, uint4 pat,
                                                  unsigned char* __restrict__ tail, size_t ntail) {
  const size_t stride = (size_t)gridDim.x * blockDim.x;
  for (size_t i = (size_t)blockIdx.x * blockDim.x + threadIdx.x; i < n16; i += stride) dst[i] = pat;
  if (blockIdx.x == 0)
    for (size_t i = threadIdx.x; i < ntail; i += blockDim.x) tail[i] = skl_pat_byte(pat, (unsigned)i);
}
// generic element size: byte-wise, the pattern staged in shared memory (a
// dynamically indexed by-value array would live in local memory)
__global__ void __launch_bounds__(256) skl_fill_bytes(unsigned char* __restrict__ dst, size_t n,
                                                      FillPattern p, int elt) {
  __shared__ unsigned char pb[64];
  if (threadIdx.x == 0) {
#pragma unroll
    for (int k = 0; k < 64; ++k) pb[k] = p.b[k];  // constant indices: read from the parameter space
  }
  __syncthreads();
  const size_t stride = (size_t)gridDim.x * blockDim.x;
  for (size_t i = (size_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride)
    dst[i] = pb[i % (size_t)elt];
}

void launch_fill(Ctx* ctx, int g, void* dst, size_t bytes, const void* value, size_t elt) {
  if (elt == 0 || elt > 64) fail(SKL_ERR_TYPE, "fill: element size must be 1..64 bytes");
  FillPattern p;
  std::memcpy(p.b, value, elt);
  Device& D = ctx->D(g);
  ctx->set_device(g);
  const unsigned grid = (unsigned)std::max<size_t>(1, std::min<size_t>((bytes / 16 + 255) / 256, (size_t)D.sm_count * 8));
  if (16 % elt == 0 && ((uintptr_t)dst & 15u) == 0) {
    uint4 pat;
    unsigned char* pb = (unsigned char*)&pat;
    for (int i = 0; i < 16; ++i) pb[i] = p.b[(size_t)i % elt];
    const size_t n16 = bytes / 16;
    skl_fill16<<<grid, 256, 0, D.stream>>>((uint4*)dst, n16, pat, (unsigned char*)dst + n16 * 16,
                                           bytes - n16 * 16);
  } else {
    skl_fill_bytes<<<grid, 256, 0, D.stream>>>((unsigned char*)dst, bytes, p, (int)elt);
  }
  SKL_CUDA(cudaGetLastError());
  ctx->n_launch++;
}

// ---------------------------------------------------------------- batched transfers
// One launch per destination GPU copies every segment of a redistribution plan
// into it (one process, several devices: same-GPU copies, or loads from a peer
// GPU's memory over NVLink when peer access is enabled).  Replaces one
// cudaMemcpy(Peer)Async per segment: a block->copy of G parts is G-1 segments per
// device, a halo refresh 2 small ones, and the per-copy launch latency
// dominated both.  Each segment is copied in units of W bytes,
// W = 16 when source and destination share their misalignment mod 16, else the
// largest power of two both share (block parts of 4-byte elements: 8 or 4);
// the unaligned head and tail (< 16 bytes) go bytewise.  The segments' bodies
// are laid end to end in a byte space (each padded to 16 bytes) cut into
// 32 KB chunks, one chunk per block iteration.
constexpr unsigned long long SKL_XCHB = 32768;
struct XferSegs {
  const unsigned char* src[kXferMaxSegs];
  unsigned char* dst[kXferMaxSegs];
  unsigned long long len[kXferMaxSegs];        // body bytes (a multiple of the unit)
  unsigned long long start[kXferMaxSegs + 1];  // byte-space offsets (16-byte multiples)
  unsigned char unit[kXferMaxSegs];            // 16, 8, 4 or 1
  // unaligned heads and tails (< 16 bytes each), copied bytewise
  const unsigned char* bsrc[2 * kXferMaxSegs];
  unsigned char* bdst[2 * kXferMaxSegs];
  unsigned char blen[2 * kXferMaxSegs];
  int nseg, nsmall;
};

template <class U>
__device__ __forceinline__ void skl_xfer_range(const unsigned char* s0, unsigned char* d0, unsigned long long lo,
                                               unsigned long long hi) {
  const U* __restrict__ s = (const U*)s0;
  U* __restrict__ d = (U*)d0;
  unsigned long long i = lo / sizeof(U) + threadIdx.x;
  const unsigned long long e = hi / sizeof(U);
  // four loads in flight per thread, then four stores
  for (; i + 3 * 256 < e; i += 4 * 256) {
    const U a = __ldcs(s + i), b = __ldcs(s + i + 256), c = __ldcs(s + i + 512), f = __ldcs(s + i + 768);
    __stcs(d + i, a);
    __stcs(d + i + 256, b);
    __stcs(d + i + 512, c);
    __stcs(d + i + 768, f);
  }
  for (; i < e; i += 256) __stcs(d + i, __ldcs(s + i));
}

__global__ void __launch_bounds__(256) skl_xfer_batch(const XferSegs S) {
  if (blockIdx.x == gridDim.x - 1)
    for (int q = (int)threadIdx.x; q < S.nsmall * 16; q += 256) {
      const int k = q >> 4, b = q & 15;
      if (b < S.blen[k]) S.bdst[k][b] = S.bsrc[k][b];
    }
  const unsigned long long total = S.start[S.nseg];
  for (unsigned long long c0 = (unsigned long long)blockIdx.x * SKL_XCHB; c0 < total;
       c0 += (unsigned long long)gridDim.x * SKL_XCHB) {
    const unsigned long long c1 = c0 + SKL_XCHB < total ? c0 + SKL_XCHB : total;
    int k = 0;
    while (S.start[k + 1] <= c0) ++k;  // first segment of the chunk (block-uniform)
    for (; k < S.nseg && S.start[k] < c1; ++k) {
      // chunk bounds relative to the segment (16-byte multiples), clipped to its body
      unsigned long long lo = c0 > S.start[k] ? c0 - S.start[k] : 0;
      unsigned long long hi = c1 - S.start[k];
      if (hi > S.len[k]) hi = S.len[k];
      if (lo >= hi) continue;
      switch (S.unit[k]) {
        case 16: skl_xfer_range<uint4>(S.src[k], S.dst[k], lo, hi); break;
        case 8: skl_xfer_range<uint2>(S.src[k], S.dst[k], lo, hi); break;
        case 4: skl_xfer_range<unsigned>(S.src[k], S.dst[k], lo, hi); break;
        default: skl_xfer_range<unsigned char>(S.src[k], S.dst[k], lo, hi); break;
      }
    }
  }
}

void launch_xfer_batch(Ctx* ctx, int g, const std::vector<XferSeg>& segs) {
  Device& D = ctx->D(g);
  ctx->set_device(g);
  for (size_t b = 0; b < segs.size(); b += kXferMaxSegs) {
    XferSegs S;
    S.nseg = (int)std::min<size_t>(kXferMaxSegs, segs.size() - b);
    S.nsmall = 0;
    S.start[0] = 0;
    auto small = [&](const unsigned char* src, unsigned char* dst, size_t n) {
      if (n == 0) return;
      S.bsrc[S.nsmall] = src;
      S.bdst[S.nsmall] = dst;
      S.blen[S.nsmall] = (unsigned char)n;
      S.nsmall++;
    };
    for (int k = 0; k < S.nseg; ++k) {
      const XferSeg& x = segs[b + (size_t)k];
      const unsigned char* sp = (const unsigned char*)x.src;
      unsigned char* dp = (unsigned char*)x.dst;
      // unit: the largest power of two (<= 16) dividing src - dst
      const uintptr_t diff = ((uintptr_t)sp - (uintptr_t)dp) & 15u;
      const size_t W = diff == 0 ? 16 : (diff & (0u - diff));
      const size_t head = std::min<size_t>(x.bytes, (W - (uintptr_t)dp % W) % W);
      const size_t body = (x.bytes - head) / W * W;
      small(sp, dp, head);
      if (x.bytes - head - body >= 16) fail(SKL_ERR_CUDA, "internal: transfer tail");
      small(sp + head + body, dp + head + body, x.bytes - head - body);
      S.src[k] = sp + head;
      S.dst[k] = dp + head;
      S.len[k] = body;
      S.unit[k] = (unsigned char)W;
      S.start[k + 1] = S.start[k] + (body + 15) / 16 * 16;
    }
    const unsigned long long total = S.start[S.nseg];
    if (total == 0 && S.nsmall == 0) continue;
    const unsigned grid = (unsigned)std::max<unsigned long long>(
        1, std::min<unsigned long long>((total + SKL_XCHB - 1) / SKL_XCHB, (unsigned long long)D.sm_count * 8));
    skl_xfer_batch<<<grid, 256, 0, D.stream>>>(S);
    SKL_CUDA(cudaGetLastError());
    ctx->n_launch++;
  }
}

// Device barrier of the IPC transport (ipc.cpp): lane h < world stores the
// epoch into rank h's signal slot for this rank (a system-scope release over
// NVLink: everything this GPU wrote before is visible to rank h first), then
// waits for rank h's epoch in this rank's slot h (acquire).  The grid is one
// warp; a wait longer than 60 s (globaltimer) raises the host-mapped error flag
// and returns instead of hanging the GPU (60 s: a peer may still be draining a
// deep queue of earlier work before it reaches its barrier).
struct SklSigSlots {
  unsigned long long* p[kIpcMaxRanks];
};
__global__ void __launch_bounds__(32) skl_ipc_barrier(SklSigSlots peers, int world, int rank,
                                                      unsigned long long* mine, unsigned long long epoch,
                                                      unsigned* err) {
  const int h = threadIdx.x;
  if (h >= world || h == rank) return;
  asm volatile("fence.acq_rel.sys;" ::: "memory");
  asm volatile("st.release.sys.global.u64 [%0], %1;" ::"l"(peers.p[h] + rank), "l"(epoch) : "memory");
  unsigned long long t0;
  asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t0));
  while (true) {
    unsigned long long v;
    asm volatile("ld.acquire.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(mine + h) : "memory");
    if (v >= epoch) break;
    unsigned long long t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    if (t - t0 > 60000000000ull) {
      atomicExch(err, 1u);
      break;
    }
    __nanosleep(200);
  }
}

void launch_ipc_barrier(Ctx* ctx, unsigned long long* const* peer_slots, int world, int rank,
                        unsigned long long* mine, unsigned long long epoch, unsigned* err) {
  SklSigSlots s{};
  for (int h = 0; h < world && h < kIpcMaxRanks; ++h) s.p[h] = peer_slots[h];
  Device& D = ctx->D(ctx->first_local);
  skl_ipc_barrier<<<1, 32, 0, D.stream>>>(s, world, rank, mine, epoch, err);
  SKL_CUDA(cudaGetLastError());
  ctx->n_launch++;
}

}  // namespace skl
