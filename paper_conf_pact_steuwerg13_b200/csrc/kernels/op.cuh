// op.cuh — the customising binary operator (+) of Reduce / Scan / combine
// (P:L264-278), wrapped as a functor, plus an L2-coherent element load.
struct SklOp {
  __device__ __forceinline__ SKL_T operator()(const SKL_T& a, const SKL_T& b) const {
    return SKL_FUNC(a, b);
  }
};

template <class T>
__device__ __forceinline__ T skl_ldcg(const T* p) {
  typename SklWords<T>::U u;
  if (sizeof(T) % 4 == 0) {
#pragma unroll
    for (int i = 0; i < SklWords<T>::N; ++i) u.w[i] = __ldcg((const unsigned*)p + i);
  } else {
    volatile const unsigned char* b = (volatile const unsigned char*)p;
    unsigned char* d = (unsigned char*)&u.t;
    for (int i = 0; i < (int)sizeof(T); ++i) d[i] = b[i];
  }
  return u.t;
}

