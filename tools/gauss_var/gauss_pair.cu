// Measured variant (profiles/sweeps/sweep_r02_gauss_pair.log): two outputs per call in
// packed fp32x2; needed an experimental skeleton hook (SKL_PAIR_FUNC) that was removed.
#define SKL_PAIR_FUNC gauss2
__device__ float skl_pc[2] = {-0.0f, 1.0f};
__device__ __forceinline__ unsigned long long skl_pk(float a, float b) {
  unsigned long long r;
  asm("mov.b64 %0, {%1, %2};" : "=l"(r) : "f"(a), "f"(b));
  return r;
}
__device__ __forceinline__ unsigned long long skl_fma2(unsigned long long a, unsigned long long b,
                                                       unsigned long long c) {
  unsigned long long d;
  asm("fma.rn.f32x2 %0, %1, %2, %3;" : "=l"(d) : "l"(a), "l"(b), "l"(c));
  return d;
}
#define SKL_PX(dx, dy) p[(dy) * SKL_PITCH + (dx)]
float2 gauss2(const float* p) {
  const unsigned long long NZ = skl_pk(skl_pc[0], skl_pc[0]), ONE = skl_pk(skl_pc[1], skl_pc[1]);
  unsigned long long acc = skl_pk(0.0f, 0.0f);
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.00296901679f, 0.00296901679f), skl_pk(SKL_PX(-2, -2), SKL_PX(-1, -2)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0133062098f, 0.0133062098f), skl_pk(SKL_PX(-1, -2), SKL_PX(0, -2)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0219382308f, 0.0219382308f), skl_pk(SKL_PX(0, -2), SKL_PX(1, -2)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0133062098f, 0.0133062098f), skl_pk(SKL_PX(1, -2), SKL_PX(2, -2)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.00296901679f, 0.00296901679f), skl_pk(SKL_PX(2, -2), SKL_PX(3, -2)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0133062098f, 0.0133062098f), skl_pk(SKL_PX(-2, -1), SKL_PX(-1, -1)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0596342944f, 0.0596342944f), skl_pk(SKL_PX(-1, -1), SKL_PX(0, -1)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0983203277f, 0.0983203277f), skl_pk(SKL_PX(0, -1), SKL_PX(1, -1)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0596342944f, 0.0596342944f), skl_pk(SKL_PX(1, -1), SKL_PX(2, -1)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0133062098f, 0.0133062098f), skl_pk(SKL_PX(2, -1), SKL_PX(3, -1)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0219382308f, 0.0219382308f), skl_pk(SKL_PX(-2, 0), SKL_PX(-1, 0)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0983203277f, 0.0983203277f), skl_pk(SKL_PX(-1, 0), SKL_PX(0, 0)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.162102818f, 0.162102818f), skl_pk(SKL_PX(0, 0), SKL_PX(1, 0)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0983203277f, 0.0983203277f), skl_pk(SKL_PX(1, 0), SKL_PX(2, 0)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0219382308f, 0.0219382308f), skl_pk(SKL_PX(2, 0), SKL_PX(3, 0)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0133062098f, 0.0133062098f), skl_pk(SKL_PX(-2, 1), SKL_PX(-1, 1)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0596342944f, 0.0596342944f), skl_pk(SKL_PX(-1, 1), SKL_PX(0, 1)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0983203277f, 0.0983203277f), skl_pk(SKL_PX(0, 1), SKL_PX(1, 1)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0596342944f, 0.0596342944f), skl_pk(SKL_PX(1, 1), SKL_PX(2, 1)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0133062098f, 0.0133062098f), skl_pk(SKL_PX(2, 1), SKL_PX(3, 1)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.00296901679f, 0.00296901679f), skl_pk(SKL_PX(-2, 2), SKL_PX(-1, 2)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0133062098f, 0.0133062098f), skl_pk(SKL_PX(-1, 2), SKL_PX(0, 2)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0219382308f, 0.0219382308f), skl_pk(SKL_PX(0, 2), SKL_PX(1, 2)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.0133062098f, 0.0133062098f), skl_pk(SKL_PX(1, 2), SKL_PX(2, 2)), NZ));
  acc = skl_fma2(acc, ONE, skl_fma2(skl_pk(0.00296901679f, 0.00296901679f), skl_pk(SKL_PX(2, 2), SKL_PX(3, 2)), NZ));
  float2 r;
  asm("mov.b64 {%0, %1}, %2;" : "=f"(r.x), "=f"(r.y) : "l"(acc));
  return r;
}
float gauss(const float* p) {
  float acc = 0.0f;
  acc = acc + 0.00296901679f * get(p, -2, -2);
  acc = acc + 0.0133062098f * get(p, -1, -2);
  acc = acc + 0.0219382308f * get(p, 0, -2);
  acc = acc + 0.0133062098f * get(p, 1, -2);
  acc = acc + 0.00296901679f * get(p, 2, -2);
  acc = acc + 0.0133062098f * get(p, -2, -1);
  acc = acc + 0.0596342944f * get(p, -1, -1);
  acc = acc + 0.0983203277f * get(p, 0, -1);
  acc = acc + 0.0596342944f * get(p, 1, -1);
  acc = acc + 0.0133062098f * get(p, 2, -1);
  acc = acc + 0.0219382308f * get(p, -2, 0);
  acc = acc + 0.0983203277f * get(p, -1, 0);
  acc = acc + 0.162102818f * get(p, 0, 0);
  acc = acc + 0.0983203277f * get(p, 1, 0);
  acc = acc + 0.0219382308f * get(p, 2, 0);
  acc = acc + 0.0133062098f * get(p, -2, 1);
  acc = acc + 0.0596342944f * get(p, -1, 1);
  acc = acc + 0.0983203277f * get(p, 0, 1);
  acc = acc + 0.0596342944f * get(p, 1, 1);
  acc = acc + 0.0133062098f * get(p, 2, 1);
  acc = acc + 0.00296901679f * get(p, -2, 2);
  acc = acc + 0.0133062098f * get(p, -1, 2);
  acc = acc + 0.0219382308f * get(p, 0, 2);
  acc = acc + 0.0133062098f * get(p, 1, 2);
  acc = acc + 0.00296901679f * get(p, 2, 2);
  return acc;
}
