#define SB(dx, dy) __int_as_float(0x4B000000 | (int)get(img, dx, dy))
uchar func(const uchar* img) {
  float h0 = SB(+1,-1) - SB(-1,-1);
  float h1 = SB(+1, 0) - SB(-1, 0);
  float h2 = SB(+1,+1) - SB(-1,+1);
  float v0 = SB(-1,+1) - SB(-1,-1);
  float v1 = SB( 0,+1) - SB( 0,-1);
  float v2 = SB(+1,+1) - SB(+1,-1);
  float h = fmaf(2.0f, h1, h0 + h2);
  float v = fmaf(2.0f, v1, v0 + v2);
  float k = fminf(fmaf(h, h, fmaf(v, v, 0.5f)), 65025.5f);
  float r, t;
  asm("sqrt.approx.ftz.f32 %0, %1;" : "=f"(r) : "f"(k));
  asm("add.rm.f32 %0, %1, 12582912.0;" : "=f"(t) : "f"(r));
  return (uchar)__float_as_int(t);
}
