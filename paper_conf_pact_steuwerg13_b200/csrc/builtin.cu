// builtin.cu — the one kernel that needs no customising function: filling a
// container's device parts with a value (skl_fill; used to zero the copy(+)
// image replicas of LM OSEM before every subset, reading A25).  Compiled by
// nvcc for sm_100a into libskl.so.
#include "skl_internal.h"

namespace skl {

struct FillPattern {
  unsigned char b[64];
};

// 16-byte stores of a 16-byte pattern (element size divides 16), byte tail.
__global__ void __launch_bounds__(256) skl_fill16(uint4* __restrict__ dst, size_t n16, uint4 pat,
                                                  unsigned char* __restrict__ tail, size_t ntail,
                                                  FillPattern p, int elt) {
  const size_t stride = (size_t)gridDim.x * blockDim.x;
  for (size_t i = (size_t)blockIdx.x * blockDim.x + threadIdx.x; i < n16; i += stride) dst[i] = pat;
  if (blockIdx.x == 0)
    for (size_t i = threadIdx.x; i < ntail; i += blockDim.x) tail[i] = p.b[(n16 * 16 + i) % (size_t)elt];
}
// generic element size: byte-wise
__global__ void __launch_bounds__(256) skl_fill_bytes(unsigned char* __restrict__ dst, size_t n,
                                                      FillPattern p, int elt) {
  const size_t stride = (size_t)gridDim.x * blockDim.x;
  for (size_t i = (size_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride)
    dst[i] = p.b[i % (size_t)elt];
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
                                           bytes - n16 * 16, p, (int)elt);
  } else {
    skl_fill_bytes<<<grid, 256, 0, D.stream>>>((unsigned char*)dst, bytes, p, (int)elt);
  }
  SKL_CUDA(cudaGetLastError());
  ctx->n_launch++;
}

}  // namespace skl
