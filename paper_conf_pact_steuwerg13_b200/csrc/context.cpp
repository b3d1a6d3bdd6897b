// context.cpp — device context and communication (SURVEY §1 layers B1, comm).
//
// SkelCL::init() makes every GPU available; skeletons then run "on all
// GPUs available in the system".  B200-native plumbing:
//  * one CUDA stream per (logical) device; stream-ordered memory pools
//    (cudaMallocAsync) with the release threshold raised so steady-state
//    allocations are free;
//  * single process, several devices: device-to-device copies
//    (cudaMemcpyPeerAsync over NVLink when the physical GPUs differ);
//  * one process per GPU (torchrun): NCCL grouped send/recv of the same
//    canonical transfer list on every rank (libnccl.so.2 via dlopen).
// The paper moves data between GPUs "via the CPU" in plain OpenCL (P:L119-121,
// P:L228-231); nothing here stages through the host.
#include <dlfcn.h>

#include <cstdio>

#include <cstdlib>

#include "skl_internal.h"

namespace skl {

static thread_local std::string g_last_error;
const char* last_error_cstr() { return g_last_error.c_str(); }
void set_last_error(const std::string& s) { g_last_error = s; }

void fail(int code, const std::string& msg) { throw Error(code, msg); }

void cuda_check(cudaError_t e, const char* what) {
  if (e == cudaSuccess) return;
  // the runtime also keeps the error as its per-thread "last error": clear it,
  // or a later cudaGetLastError() (after a launch) would report this failure
  // again (non-sticky errors such as a failed allocation leave the context usable)
  (void)cudaGetLastError();
  const int code = (e == cudaErrorMemoryAllocation) ? SKL_ERR_OOM : SKL_ERR_CUDA;
  fail(code, std::string(what) + ": " + cudaGetErrorName(e) + " (" + cudaGetErrorString(e) + ")");
}

const TypeInfo& Ctx::type(int t) const {
  if (t < 0 || (size_t)t >= types.size() || types[(size_t)t].size == 0)
    fail(SKL_ERR_TYPE, "unknown element type " + std::to_string(t));
  return types[(size_t)t];
}

void Ctx::set_device(int g) {
  if (offline) fail(SKL_ERR_CUDA, "offline context (skl_init_offline) has no devices");
  SKL_CUDA(cudaSetDevice(D(g).phys));
}

// Environment defaults: SKL_BLOCK_THREADS (work-group size,
// P:L470), SKL_DEBUG_BOUNDS (A21); skl_set_option overrides both.  SKL_CACHE_DIR
// is read by the compiler (on-disk cubin cache).
static void apply_env(Ctx* c) {
  if (const char* v = std::getenv("SKL_BLOCK_THREADS")) {
    const long b = std::strtol(v, nullptr, 10);
    if (b >= 64 && b <= 1024 && b % 32 == 0) c->block_threads = (int)b;
  }
  if (const char* v = std::getenv("SKL_DEBUG_BOUNDS")) c->debug_bounds = std::strtol(v, nullptr, 10) != 0;
}

static void init_types(Ctx* c) {
  apply_env(c);
  c->types.resize(12);
  c->types[SKL_VOID] = {"void", 0, 1, ""};
  c->types[SKL_U8] = {"unsigned char", 1, 1, ""};
  c->types[SKL_I8] = {"signed char", 1, 1, ""};
  c->types[SKL_I32] = {"int", 4, 4, ""};
  c->types[SKL_U32] = {"unsigned int", 4, 4, ""};
  c->types[SKL_F32] = {"float", 4, 4, ""};
  c->types[SKL_F64] = {"double", 8, 8, ""};
  c->types[SKL_F32X2] = {"float2", 8, 8, ""};
  c->types[SKL_I64] = {"long long", 8, 8, ""};
  c->types[SKL_U64] = {"unsigned long long", 8, 8, ""};
  c->types[SKL_I16] = {"short", 2, 2, ""};
  c->types[SKL_U16] = {"unsigned short", 2, 2, ""};
}

static void init_device(Ctx* c, Device& d) {
  SKL_CUDA(cudaSetDevice(d.phys));
  SKL_CUDA(cudaStreamCreateWithFlags(&d.own, cudaStreamNonBlocking));
  d.stream = d.own;
  SKL_CUDA(cudaEventCreateWithFlags(&d.ev, cudaEventDisableTiming));
  SKL_CUDA(cudaStreamCreateWithFlags(&d.h2d, cudaStreamNonBlocking));
  SKL_CUDA(cudaStreamCreateWithFlags(&d.d2h, cudaStreamNonBlocking));
  SKL_CUDA(cudaDeviceGetAttribute(&d.sm_count, cudaDevAttrMultiProcessorCount, d.phys));
  cudaMemPool_t pool;
  SKL_CUDA(cudaDeviceGetDefaultMemPool(&pool, d.phys));
  uint64_t thr = UINT64_MAX;
  SKL_CUDA(cudaMemPoolSetAttribute(pool, cudaMemPoolAttrReleaseThreshold, &thr));
  (void)c;
}

Ctx* ctx_create_local(int ndev, const int* devices) {
  int nvis = 0;
  cudaError_t e = cudaGetDeviceCount(&nvis);
  if (e != cudaSuccess || nvis <= 0)
    fail(SKL_ERR_CUDA, std::string("no CUDA device available: ") + cudaGetErrorString(e));
  auto* c = new Ctx();
  init_types(c);
  c->G = ndev > 0 ? ndev : nvis;
  c->first_local = 0;
  c->nlocal = c->G;
  c->dev.resize((size_t)c->G);
  try {
    for (int g = 0; g < c->G; ++g) {
      c->dev[(size_t)g].global = g;
      c->dev[(size_t)g].phys = devices ? devices[g] : g % nvis;
      if (c->dev[(size_t)g].phys < 0 || c->dev[(size_t)g].phys >= nvis)
        fail(SKL_ERR_INVALID_ARG, "device ordinal out of range");
      init_device(c, c->dev[(size_t)g]);
    }
    // peer access between distinct physical GPUs (NVLink / NVSwitch).  Two
    // grants are needed for a kernel on GPU a to load/store GPU b's buffers:
    // cudaDeviceEnablePeerAccess covers cudaMalloc memory (and the caller's
    // allocator, e.g. torch's), and cudaMemPoolSetAccess gives a access to b's
    // default stream-ordered pool, where device_alloc places every part and
    // scratch buffer.  peer_ok[a][b] is set only when both succeed; otherwise
    // the moves from b into a use the copy engines (cudaMemcpyPeerAsync) and the
    // fused peer kernels (halo push, copy(+)->block fold, Reduce fold) stay off.
    c->peer_ok.assign((size_t)c->G, std::vector<char>((size_t)c->G, 0));
    std::map<std::pair<int, int>, char> phys_ok;  // (a.phys, b.phys) -> granted
    for (auto& a : c->dev)
      for (auto& b : c->dev) {
        char& ok = c->peer_ok[(size_t)a.global][(size_t)b.global];
        if (a.phys == b.phys) {
          ok = 1;
          continue;
        }
        auto key = std::make_pair(a.phys, b.phys);
        auto it = phys_ok.find(key);
        if (it != phys_ok.end()) {
          ok = it->second;
          continue;
        }
        int can = 0;
        cudaDeviceCanAccessPeer(&can, a.phys, b.phys);
        if (can) {
          cudaSetDevice(a.phys);
          cudaError_t pe = cudaDeviceEnablePeerAccess(b.phys, 0);
          if (pe == cudaErrorPeerAccessAlreadyEnabled) pe = cudaSuccess;
          if (pe == cudaSuccess) {
            cudaMemPool_t bpool;
            pe = cudaDeviceGetDefaultMemPool(&bpool, b.phys);
            if (pe == cudaSuccess) {
              cudaMemAccessDesc desc{};
              desc.location.type = cudaMemLocationTypeDevice;
              desc.location.id = a.phys;
              desc.flags = cudaMemAccessFlagsProtReadWrite;
              pe = cudaMemPoolSetAccess(bpool, &desc, 1);
            }
          }
          if (pe != cudaSuccess) cudaGetLastError();
          ok = pe == cudaSuccess;
        }
        phys_ok[key] = ok;
      }
  } catch (...) {
    delete c;
    throw;
  }
  return c;
}

Ctx* ctx_create_dist(int rank, int world, int cuda_device, const void* nccl_id) {
  int nvis = 0;
  cudaError_t e = cudaGetDeviceCount(&nvis);
  if (e != cudaSuccess || nvis <= 0)
    fail(SKL_ERR_CUDA, std::string("no CUDA device available: ") + cudaGetErrorString(e));
  if (world < 1 || rank < 0 || rank >= world) fail(SKL_ERR_INVALID_ARG, "bad rank/world");
  auto* c = new Ctx();
  init_types(c);
  c->G = world;
  // SKL_DIST_FORCE=1: the multi-process code path and its transport even for
  // one rank, so the transport's setup, group calls and teardown (NCCL's
  // included, which refuses two ranks on one GPU) run on a one-GPU box
  const char* force = std::getenv("SKL_DIST_FORCE");
  c->dist_mode = world > 1 || (force && std::string(force) == "1");
  c->rank = rank;
  c->world = world;
  c->first_local = rank;
  c->nlocal = 1;
  c->dev.resize(1);
  c->dev[0].global = rank;
  c->dev[0].phys = cuda_device;
  try {
    init_device(c, c->dev[0]);
    if (c->dist_mode) nccl_init(c, nccl_id);
  } catch (...) {
    delete c;
    throw;
  }
  return c;
}

Ctx* ctx_create_offline() {
  auto* c = new Ctx();
  init_types(c);
  c->offline = true;
  c->G = 1;
  c->nlocal = 0;
  return c;
}

void ctx_destroy(Ctx* c) {
  for (auto& d : c->dev) {
    cudaSetDevice(d.phys);
    cudaStreamSynchronize(d.stream);
    cudaStreamSynchronize(d.own);
    if (d.h2d) cudaStreamSynchronize(d.h2d);
    if (d.d2h) cudaStreamSynchronize(d.d2h);
  }
  while (!c->skels.empty()) skel_destroy(*c->skels.begin());
  while (!c->conts.empty()) cont_destroy(*c->conts.begin());
  for (auto& kv : c->programs)
    if (kv.second) {
      // cudaLibraryUnload is safe after the streams drained
      extern void program_unload(Program*);
      program_unload(kv.second.get());
    }
  if (c->nccl_comm || c->shm_comm || c->ipc) nccl_destroy(c);
  for (auto& d : c->dev) {
    cudaSetDevice(d.phys);
    if (d.ev) cudaEventDestroy(d.ev);
    for (cudaEvent_t e : d.ev_pool) cudaEventDestroy(e);
    if (d.h2d) cudaStreamDestroy(d.h2d);
    if (d.d2h) cudaStreamDestroy(d.d2h);
    if (d.own) cudaStreamDestroy(d.own);
  }
  if (c->cap_fork) cudaEventDestroy(c->cap_fork);
  for (cudaEvent_t e : c->cap_join)
    if (e) cudaEventDestroy(e);
  delete c;
}

void* device_alloc(Ctx* ctx, int g, size_t bytes) {
  if (bytes == 0) bytes = 16;
  ctx->set_device(g);
  void* p = nullptr;
  // one process per GPU over NVLink: every buffer a peer may read or write
  // lives in the IPC heap (ipc.cpp); it takes precedence over a caller's allocator
  if (ctx->ipc) return ipc_alloc(ctx, bytes);
  if (ctx->user_alloc) {
    // caller's allocator (e.g. torch's caching allocator), stream-ordered on
    // this device's stream
    p = ctx->user_alloc(bytes, ctx->D(g).phys, (void*)ctx->D(g).stream, ctx->alloc_user);
    if (!p) fail(SKL_ERR_OOM, "user allocator returned NULL for " + std::to_string(bytes) + " bytes");
    return p;
  }
  SKL_CUDA(cudaMallocAsync(&p, bytes, ctx->D(g).stream));
  return p;
}
void device_free(Ctx* ctx, int g, void* p) {
  if (!p) return;
  ctx->set_device(g);
  if (ctx->ipc) {
    // the range is reused by later allocations, whose work is ordered after
    // this stream's; peers read it only between device barriers
    ipc_free(ctx, p);
    return;
  }
  if (ctx->user_free) {
    // the block may be reused at once on this stream: work other devices'
    // streams queued on it (peer copies) must be ordered before that reuse
    if (ctx->nlocal > 1) barrier_streams(ctx);
    ctx->user_free(p, ctx->D(g).phys, (void*)ctx->D(g).stream, ctx->alloc_user);
    return;
  }
  SKL_CUDA(cudaFreeAsync(p, ctx->D(g).stream));
}

// Reusable events (a stream wait captures the event's state when it is issued,
// so an event can be re-recorded as soon as the waits on it are enqueued).
cudaEvent_t event_get(Ctx* ctx, int g) {
  Device& d = ctx->D(g);
  if (!d.ev_pool.empty()) {
    cudaEvent_t e = d.ev_pool.back();
    d.ev_pool.pop_back();
    return e;
  }
  ctx->set_device(g);
  cudaEvent_t e = nullptr;
  SKL_CUDA(cudaEventCreateWithFlags(&e, cudaEventDisableTiming));
  return e;
}
void event_put(Ctx* ctx, int g, cudaEvent_t e) {
  if (e) ctx->D(g).ev_pool.push_back(e);
}

// Every local stream waits for the work already queued on every other local
// stream: orders a multi-device exchange after its producers and before its
// consumers (G <= 8, so at most 64 event waits).
void barrier_streams(Ctx* ctx) {
  if (ctx->nlocal <= 1) return;
  // devices that share a stream (e.g. logical devices handed one caller
  // stream) are already ordered with each other
  bool one_stream = true;
  for (auto& d : ctx->dev) one_stream = one_stream && d.stream == ctx->dev[0].stream;
  if (one_stream) return;
  for (auto& d : ctx->dev) {
    SKL_CUDA(cudaSetDevice(d.phys));
    SKL_CUDA(cudaEventRecord(d.ev, d.stream));
  }
  for (auto& a : ctx->dev) {
    SKL_CUDA(cudaSetDevice(a.phys));
    for (auto& b : ctx->dev)
      if (&a != &b && a.stream != b.stream) SKL_CUDA(cudaStreamWaitEvent(a.stream, b.ev, 0));
  }
}

}  // namespace skl
