uchar func(const uchar* img) {
  float h0 = (float)get(img,+1,-1) - (float)get(img,-1,-1);
  float h1 = (float)get(img,+1, 0) - (float)get(img,-1, 0);
  float h2 = (float)get(img,+1,+1) - (float)get(img,-1,+1);
  float v0 = (float)get(img,-1,+1) - (float)get(img,-1,-1);
  float v1 = (float)get(img, 0,+1) - (float)get(img, 0,-1);
  float v2 = (float)get(img,+1,+1) - (float)get(img,+1,-1);
  float h = fmaf(2.0f, h1, h0 + h2);
  float v = fmaf(2.0f, v1, v0 + v2);
  float k = fmaf(h, h, fmaf(v, v, 0.5f));
  float r;
  asm("sqrt.approx.ftz.f32 %0, %1;" : "=f"(r) : "f"(k));
  unsigned q = __float2uint_rz(r);
  return (uchar)(q > 255u ? 255u : q);
}
