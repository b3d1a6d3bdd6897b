uchar func(const uchar* img) {
  int h0 = get(img,+1,-1) - get(img,-1,-1);
  int h1 = get(img,+1, 0) - get(img,-1, 0);
  int h2 = get(img,+1,+1) - get(img,-1,+1);
  int v0 = get(img,-1,+1) - get(img,-1,-1);
  int v1 = get(img, 0,+1) - get(img, 0,-1);
  int v2 = get(img,+1,+1) - get(img,+1,-1);
  int h = h0 + 2 * h1 + h2, v = v0 + 2 * v1 + v2;
  const int m = h * h + (v * v + 0x4B000000);
  float k = fminf(__int_as_float(m) - 8388607.5f, 65025.5f);
  float r, t;
  asm("sqrt.approx.ftz.f32 %0, %1;" : "=f"(r) : "f"(k));
  asm("add.rm.f32 %0, %1, 12582912.0;" : "=f"(t) : "f"(r));
  return (uchar)__float_as_int(t);
}