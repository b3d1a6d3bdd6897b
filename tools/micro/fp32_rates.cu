// fp32_rates.cu — FP32 pipe throughput on sm_100a (B200): FADD / FMUL / FFMA,
// register vs immediate operand, and the packed f32x2 forms (FADD2 / FMUL2 /
// FFMA2).  Each thread runs 8 independent chains; ops per SM per cycle come from
// %clock64 around the loop in every block (max over a block's warps), so the
// number does not depend on the clock the GPU happens to run at.
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o fp32_rates fp32_rates.cu
#include <cstdio>
#include <cuda_runtime.h>

#define ITERS 4096
#define CH 8

__device__ __forceinline__ unsigned long long f2u(float2 v) { return *(unsigned long long*)&v; }
__device__ __forceinline__ float2 u2f(unsigned long long v) { return *(float2*)&v; }

template <int MODE>
__global__ void k(float* out, float a, float b, unsigned long long* cyc) {
  float x[CH], y[CH];
  unsigned long long p[CH], q[CH];
#pragma unroll
  for (int c = 0; c < CH; ++c) {
    x[c] = threadIdx.x * 1e-3f + c;
    p[c] = f2u(make_float2(x[c], x[c] + 0.5f));
    y[c] = x[c] * 0.5f;
    q[c] = f2u(make_float2(y[c], y[c] + 0.25f));
  }
  const unsigned long long pa = f2u(make_float2(a, a)), pb = f2u(make_float2(b, b));
  __syncthreads();
  long long t0 = clock64();
  for (int i = 0; i < ITERS; ++i) {
#pragma unroll
    for (int c = 0; c < CH; ++c) {
      if (MODE == 0) asm volatile("add.rn.f32 %0, %0, %1;" : "+f"(x[c]) : "f"(a));           // FADD reg
      if (MODE == 1) asm volatile("mul.rn.f32 %0, %0, 0f3F800001;" : "+f"(x[c]));           // FMUL imm
      if (MODE == 2) asm volatile("mul.rn.f32 %0, %0, %1;" : "+f"(x[c]) : "f"(a));           // FMUL reg
      if (MODE == 3) asm volatile("fma.rn.f32 %0, %0, %1, %2;" : "+f"(x[c]) : "f"(a), "f"(b));  // FFMA reg
      if (MODE == 4) asm volatile("add.rn.f32x2 %0, %0, %1;" : "+l"(p[c]) : "l"(pa));        // FADD2
      if (MODE == 5) asm volatile("mul.rn.f32x2 %0, %0, %1;" : "+l"(p[c]) : "l"(pa));        // FMUL2
      if (MODE == 6) asm volatile("fma.rn.f32x2 %0, %0, %1, %2;" : "+l"(p[c]) : "l"(pa), "l"(pb));  // FFMA2
      if (MODE == 7) {  // Gaussian pattern: acc = acc + w * v  (FMUL imm + FADD reg)
        asm volatile("mul.rn.f32 %0, %0, 0f3F800001;" : "+f"(y[c]));
        asm volatile("add.rn.f32 %0, %0, %1;" : "+f"(x[c]) : "f"(y[c]));
      }
      if (MODE == 8) {  // the same on f32x2
        asm volatile("mul.rn.f32x2 %0, %0, %1;" : "+l"(q[c]) : "l"(pa));
        asm volatile("add.rn.f32x2 %0, %0, %1;" : "+l"(p[c]) : "l"(q[c]));
      }
    }
  }
  long long t1 = clock64();
  float s = 0.f;
#pragma unroll
  for (int c = 0; c < CH; ++c) s += x[c] + y[c] + u2f(p[c]).x + u2f(p[c]).y + u2f(q[c]).x;
  out[blockIdx.x * blockDim.x + threadIdx.x] = s;
  if ((threadIdx.x & 31) == 0) atomicMax(&cyc[blockIdx.x], (unsigned long long)(t1 - t0));
}

template <int MODE>
void run(const char* name, int lanes_per_inst, int insts_per_chain_step) {
  int sms;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  const int threads = 1024, blocks = sms;  // one 1024-thread block per SM (32 warps)
  float* out;
  unsigned long long* cyc;
  cudaMalloc(&out, sizeof(float) * threads * blocks);
  cudaMalloc(&cyc, sizeof(unsigned long long) * blocks);
  cudaMemset(cyc, 0, sizeof(unsigned long long) * blocks);
  k<MODE><<<blocks, threads>>>(out, 1.0000001f, 1e-7f, cyc);
  cudaMemset(cyc, 0, sizeof(unsigned long long) * blocks);
  cudaEvent_t e0, e1;
  cudaEventCreate(&e0);
  cudaEventCreate(&e1);
  cudaEventRecord(e0);
  k<MODE><<<blocks, threads>>>(out, 1.0000001f, 1e-7f, cyc);
  cudaEventRecord(e1);
  cudaEventSynchronize(e1);
  float ms;
  cudaEventElapsedTime(&ms, e0, e1);
  unsigned long long h[1024];
  cudaMemcpy(h, cyc, sizeof(unsigned long long) * blocks, cudaMemcpyDeviceToHost);
  double mx = 0;
  for (int i = 0; i < blocks; ++i) mx = h[i] > mx ? h[i] : mx;
  const double warp_insts = (double)threads / 32 * ITERS * CH * insts_per_chain_step;  // per SM
  const double lane_ops = warp_insts * 32 * lanes_per_inst;
  printf("%-34s warp-inst/clk/SM %6.3f  fp32 lane-ops/clk/SM %7.2f  (%.3f ms, %.0f cycles, %.1f GHz eff)\n", name,
         warp_insts / mx, lane_ops / mx, ms, mx, mx / (ms * 1e6));
  cudaFree(out);
  cudaFree(cyc);
}

int main() {
  run<0>("FADD reg", 1, 1);
  run<1>("FMUL imm", 1, 1);
  run<2>("FMUL reg", 1, 1);
  run<3>("FFMA reg (2 ops/lane)", 2, 1);
  run<4>("FADD2 f32x2", 2, 1);
  run<5>("FMUL2 f32x2", 2, 1);
  run<6>("FFMA2 f32x2 (4 ops/lane)", 4, 1);
  run<7>("FMUL imm + FADD reg (gauss)", 1, 2);
  run<8>("FMUL2 + FADD2 (gauss x2)", 2, 2);
  return 0;
}
