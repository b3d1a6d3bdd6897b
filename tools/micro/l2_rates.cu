// l2_rates.cu — L2 throughput for the LM OSEM access pattern on sm_100a (B200):
// random 16-byte gathers (ld.global.nc.v4.f32) and random 16-byte vector atomics
// (red.global.add.v4.f32), and the 4-byte forms, into a buffer of the LM OSEM
// image size (150^3 floats = 13.5 MB, L2-resident).  Reports L2 requests/s (one
// request = one 32-byte sector here: every access is 16-byte aligned).
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o l2_rates l2_rates.cu
#include <cstdio>
#include <cuda_runtime.h>

#define N_GROUPS (150 * 150 * 150 / 4)

__device__ __forceinline__ unsigned hash(unsigned x) {
  x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16;
  return x;
}

template <int MODE>
__global__ void k(float* buf, int iters, float* sink) {
  const unsigned t = blockIdx.x * blockDim.x + threadIdx.x;
  float acc = 0.f;
  unsigned s = hash(t * 0x9E3779B9u + 1u);
  for (int i = 0; i < iters; ++i) {
    s = hash(s);
    const unsigned g = s % N_GROUPS;
    float* p = buf + 4 * (size_t)g;
    if (MODE == 0) {
      float4 v;
      asm volatile("ld.global.nc.v4.f32 {%0,%1,%2,%3}, [%4];" : "=f"(v.x), "=f"(v.y), "=f"(v.z), "=f"(v.w) : "l"(p));
      acc += v.x + v.w;
    } else if (MODE == 1) {
      asm volatile("red.global.add.v4.f32 [%0], {%1,%1,%1,%1};" ::"l"(p), "f"(1e-9f) : "memory");
    } else if (MODE == 2) {
      float v;
      asm volatile("ld.global.nc.f32 %0, [%1];" : "=f"(v) : "l"(p + (s >> 30)));
      acc += v;
    } else {
      asm volatile("red.global.add.f32 [%0], %1;" ::"l"(p + (s >> 30)), "f"(1e-9f) : "memory");
    }
  }
  if (acc == 12345.f) sink[0] = acc;
}

template <int MODE>
void run(const char* name) {
  int sms;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  float *buf, *sink;
  cudaMalloc(&buf, sizeof(float) * 4 * (size_t)N_GROUPS);
  cudaMalloc(&sink, 4);
  cudaMemset(buf, 0, sizeof(float) * 4 * (size_t)N_GROUPS);
  const int threads = 256, blocks = sms * 8, iters = 2048;
  k<MODE><<<blocks, threads>>>(buf, 64, sink);
  cudaEvent_t e0, e1;
  cudaEventCreate(&e0);
  cudaEventCreate(&e1);
  cudaEventRecord(e0);
  k<MODE><<<blocks, threads>>>(buf, iters, sink);
  cudaEventRecord(e1);
  cudaEventSynchronize(e1);
  float ms;
  cudaEventElapsedTime(&ms, e0, e1);
  const double ops = (double)blocks * threads * iters;
  printf("%-28s %.3f ms  %.3e requests/s  (%.1f GB/s of 32-byte sectors)\n", name, ms, ops / (ms * 1e-3),
         ops * 32 / (ms * 1e-3) / 1e9);
  cudaFree(buf);
  cudaFree(sink);
}

int main() {
  run<0>("gather ld.v4 16 B random");
  run<1>("red.add.v4.f32 16 B random");
  run<2>("gather ld 4 B random");
  run<3>("red.add.f32 4 B random");
  return 0;
}
