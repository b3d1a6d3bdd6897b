// common.cuh — device helpers shared by the skeleton kernel templates.
// Appended after the user's source; everything here is sm_100a device code.
#define SKL_FULL 0xffffffffu

typedef unsigned long long skl_u64;

// 128-bit streaming accesses (Guideline 13): loads bypass L1 allocation and
// stores are evict-first, the right policy for read-once / write-once streams.
__device__ __forceinline__ uint4 skl_ld16(const void* p) {
  uint4 r;
  // not volatile: a read-only load the compiler may hoist / batch (MLP)
  asm("ld.global.nc.L1::no_allocate.v4.u32 {%0,%1,%2,%3}, [%4];"
               : "=r"(r.x), "=r"(r.y), "=r"(r.z), "=r"(r.w) : "l"(p));
  return r;
}
__device__ __forceinline__ void skl_st16(void* p, uint4 v) {
  asm volatile("st.global.cs.v4.u32 [%0], {%1,%2,%3,%4};" ::"l"(p), "r"(v.x), "r"(v.y), "r"(v.z),
               "r"(v.w) : "memory");
}

// V elements of T viewed as 16-byte words (V*sizeof(T) is a multiple of 16).
template <class T, int V>
union SklChunk {
  T e[V];
  uint4 q[(V * sizeof(T) + 15) / 16];
  __device__ SklChunk() {}
};

// acquire / release on the decoupled-lookback status words
__device__ __forceinline__ unsigned skl_ld_acquire(const unsigned* p) {
  unsigned v;
  asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void skl_st_release(unsigned* p, unsigned v) {
  asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}

// Element type moved as 32-bit words through shuffles (any trivially copyable T).
template <class T>
struct SklWords {
  enum { N = (sizeof(T) + 3) / 4 };
  union U {
    T t;
    unsigned w[N];
    __device__ U() {}
  };
};
template <class T>
__device__ __forceinline__ T skl_shfl_down(T v, int s) {
  typename SklWords<T>::U u;
  u.t = v;
#pragma unroll
  for (int i = 0; i < SklWords<T>::N; ++i) u.w[i] = __shfl_down_sync(SKL_FULL, u.w[i], s);
  return u.t;
}
template <class T>
__device__ __forceinline__ T skl_shfl_up(T v, int s) {
  typename SklWords<T>::U u;
  u.t = v;
#pragma unroll
  for (int i = 0; i < SklWords<T>::N; ++i) u.w[i] = __shfl_up_sync(SKL_FULL, u.w[i], s);
  return u.t;
}
template <class T>
__device__ __forceinline__ T skl_shfl(T v, int lane) {
  typename SklWords<T>::U u;
  u.t = v;
#pragma unroll
  for (int i = 0; i < SklWords<T>::N; ++i) u.w[i] = __shfl_sync(SKL_FULL, u.w[i], lane);
  return u.t;
}

// Order-preserving warp fold of the first `nv` lanes (nv >= 1): lane 0 returns
// v_0 (+) v_1 (+) ... (+) v_{nv-1}.  The left operand always has the lower lane,
// and invalid lanes are skipped, never padded with an identity ((+)
// is only associative; reading A10).
template <class T, class F>
__device__ __forceinline__ T skl_warp_fold(T v, int nv, F op) {
  const int lane = threadIdx.x & 31;
#pragma unroll
  for (int s = 1; s < 32; s <<= 1) {
    T o = skl_shfl_down(v, s);
    if (lane + s < nv) v = op(v, o);
  }
  return v;
}
