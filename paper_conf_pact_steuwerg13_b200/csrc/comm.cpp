// comm.cpp — execution of inter-device transfer lists.
//
// A redistribution is planned once on the host (plan.cpp) as a
// canonical list of (src device, dst device, unit range) moves.  One process:
// every move is a stream-ordered device-to-device copy on the destination's
// stream (peer copy over NVLink between physical GPUs).  One process per GPU:
// every rank walks the same list inside one ncclGroupStart/End and posts the
// ncclSend / ncclRecv halves that touch it, so matching pairs are issued in the
// same order on both sides (NCCL matches p2p operations per peer in order).
#include <dlfcn.h>
#include <fcntl.h>
#include <nccl.h>
#include <sys/mman.h>
#include <unistd.h>

#include <atomic>
#include <chrono>
#include <cstdlib>
#include <mutex>
#include <random>
#include <thread>

#include "skl_internal.h"

namespace skl {

namespace {
struct NcclApi {
  void* h = nullptr;
  decltype(&ncclGetUniqueId) getUniqueId = nullptr;
  decltype(&ncclCommInitRank) commInitRank = nullptr;
  decltype(&ncclCommDestroy) commDestroy = nullptr;
  decltype(&ncclGroupStart) groupStart = nullptr;
  decltype(&ncclGroupEnd) groupEnd = nullptr;
  decltype(&ncclSend) send = nullptr;
  decltype(&ncclRecv) recv = nullptr;
  decltype(&ncclGetErrorString) errstr = nullptr;
  decltype(&ncclCommGetAsyncError) asyncError = nullptr;
};
NcclApi* nccl() {
  static NcclApi a;
  static std::once_flag once;
  std::call_once(once, [] {
    // the copy already in the process first (torch's bundled NCCL when torch was
    // imported): one NCCL build per process, never two side by side
    a.h = dlopen("libnccl.so.2", RTLD_NOW | RTLD_NOLOAD);
    const char* names[] = {"libnccl.so.2", "/usr/lib/x86_64-linux-gnu/libnccl.so.2", "libnccl.so"};
    for (const char* n : names) {
      if (a.h) break;
      a.h = dlopen(n, RTLD_NOW | RTLD_GLOBAL);
    }
    if (!a.h) return;
    a.getUniqueId = (decltype(a.getUniqueId))dlsym(a.h, "ncclGetUniqueId");
    a.commInitRank = (decltype(a.commInitRank))dlsym(a.h, "ncclCommInitRank");
    a.commDestroy = (decltype(a.commDestroy))dlsym(a.h, "ncclCommDestroy");
    a.groupStart = (decltype(a.groupStart))dlsym(a.h, "ncclGroupStart");
    a.groupEnd = (decltype(a.groupEnd))dlsym(a.h, "ncclGroupEnd");
    a.send = (decltype(a.send))dlsym(a.h, "ncclSend");
    a.recv = (decltype(a.recv))dlsym(a.h, "ncclRecv");
    a.errstr = (decltype(a.errstr))dlsym(a.h, "ncclGetErrorString");
    a.asyncError = (decltype(a.asyncError))dlsym(a.h, "ncclCommGetAsyncError");
  });
  if (!a.h || !a.commInitRank || !a.send || !a.recv)
    fail(SKL_ERR_UNSUPPORTED, "NCCL (libnccl.so.2) could not be loaded");
  return &a;
}
void nccl_check(ncclResult_t r, const char* what) {
  if (r == ncclSuccess) return;
  NcclApi* a = nccl();
  fail(SKL_ERR_NCCL, std::string(what) + ": " + (a->errstr ? a->errstr(r) : "NCCL error"));
}
}  // namespace

// ---- host shared-memory loopback transport (SKL_COMM=shm) ------------------
// Test transport for the one-process-per-GPU mode with several processes on ONE
// GPU (NCCL refuses two ranks on one device; SURVEY §4 T3 "loopback backend").
// Every rank walks the same canonical transfer list in the same order: a send
// copies the units device -> a POSIX shared-memory object and publishes a
// per-(src, dst) sequence number; the matching receive waits for it and copies
// shared memory -> device.  Sends never block, so the list order cannot
// deadlock.  Slow (two host copies), correct, and never used unless asked for.
namespace {
struct ShmComm {
  std::string name;
  int rank = 0, world = 1;
  std::atomic<unsigned long long>* seq = nullptr;  // world x world published counters
  size_t ctl_bytes = 0;
  std::vector<unsigned long long> sent, recvd;     // this rank's counters per pair
};
bool shm_mode() {
  const char* v = std::getenv("SKL_COMM");
  return v && std::string(v) == "shm";
}
std::string shm_data_name(const ShmComm& c, int src, int dst, unsigned long long k) {
  return c.name + "_" + std::to_string(src) + "_" + std::to_string(dst) + "_" + std::to_string(k);
}
void shm_send(Ctx* ctx, ShmComm& c, const void* dptr, size_t bytes, int dst) {
  Device& L = ctx->D(ctx->first_local);
  const size_t pair = (size_t)c.rank * c.world + dst;
  const unsigned long long k = c.sent[pair]++;
  const std::string nm = shm_data_name(c, c.rank, dst, k);
  const int fd = shm_open(nm.c_str(), O_CREAT | O_RDWR | O_TRUNC, 0600);
  if (fd < 0) fail(SKL_ERR_NCCL, "shm transport: shm_open failed for " + nm);
  if (ftruncate(fd, (off_t)std::max<size_t>(bytes, 1)) != 0) {
    close(fd);
    fail(SKL_ERR_NCCL, "shm transport: ftruncate failed");
  }
  void* h = mmap(nullptr, std::max<size_t>(bytes, 1), PROT_READ | PROT_WRITE, MAP_SHARED, fd, 0);
  close(fd);
  if (h == MAP_FAILED) fail(SKL_ERR_NCCL, "shm transport: mmap failed");
  SKL_CUDA(cudaMemcpyAsync(h, dptr, bytes, cudaMemcpyDeviceToHost, L.stream));  // after its producers
  SKL_CUDA(cudaStreamSynchronize(L.stream));
  munmap(h, std::max<size_t>(bytes, 1));
  c.seq[pair].store(k + 1, std::memory_order_release);
}
void shm_recv(Ctx* ctx, ShmComm& c, void* dptr, size_t bytes, int src) {
  Device& L = ctx->D(ctx->first_local);
  const size_t pair = (size_t)src * c.world + c.rank;
  const unsigned long long k = c.recvd[pair]++;
  const auto t0 = std::chrono::steady_clock::now();
  while (c.seq[pair].load(std::memory_order_acquire) <= k) {
    if (std::chrono::steady_clock::now() - t0 > std::chrono::seconds(300))
      fail(SKL_ERR_NCCL, "shm transport: timed out waiting for rank " + std::to_string(src));
    std::this_thread::sleep_for(std::chrono::microseconds(50));
  }
  const std::string nm = shm_data_name(c, src, c.rank, k);
  const int fd = shm_open(nm.c_str(), O_RDONLY, 0600);
  if (fd < 0) fail(SKL_ERR_NCCL, "shm transport: missing " + nm);
  void* h = mmap(nullptr, std::max<size_t>(bytes, 1), PROT_READ, MAP_SHARED, fd, 0);
  close(fd);
  if (h == MAP_FAILED) fail(SKL_ERR_NCCL, "shm transport: mmap failed");
  SKL_CUDA(cudaMemcpyAsync(dptr, h, bytes, cudaMemcpyHostToDevice, L.stream));
  SKL_CUDA(cudaStreamSynchronize(L.stream));
  munmap(h, std::max<size_t>(bytes, 1));
  shm_unlink(nm.c_str());
}
void shm_init(Ctx* ctx, const void* id128) {
  auto* c = new ShmComm();
  c->name = std::string((const char*)id128, strnlen((const char*)id128, 127));
  c->rank = ctx->rank;
  c->world = ctx->world;
  c->ctl_bytes = (size_t)c->world * c->world * sizeof(unsigned long long);
  const std::string ctl = c->name + "_ctl";
  const int fd = shm_open(ctl.c_str(), O_CREAT | O_RDWR, 0600);
  if (fd < 0) {
    delete c;
    fail(SKL_ERR_NCCL, "shm transport: cannot open " + ctl);
  }
  if (ftruncate(fd, (off_t)c->ctl_bytes) != 0) {  // same size on every rank: idempotent
    close(fd);
    delete c;
    fail(SKL_ERR_NCCL, "shm transport: ftruncate failed");
  }
  void* h = mmap(nullptr, c->ctl_bytes, PROT_READ | PROT_WRITE, MAP_SHARED, fd, 0);
  close(fd);
  if (h == MAP_FAILED) {
    delete c;
    fail(SKL_ERR_NCCL, "shm transport: mmap failed");
  }
  c->seq = (std::atomic<unsigned long long>*)h;
  c->sent.assign((size_t)c->world * c->world, 0);
  c->recvd.assign((size_t)c->world * c->world, 0);
  ctx->shm_comm = c;
}
void shm_destroy(Ctx* ctx) {
  auto* c = (ShmComm*)ctx->shm_comm;
  if (!c) return;
  munmap((void*)c->seq, c->ctl_bytes);
  if (c->rank == 0) shm_unlink((c->name + "_ctl").c_str());
  delete c;
  ctx->shm_comm = nullptr;
}
}  // namespace

void nccl_get_unique_id(void* out128) {
  if (shm_mode() || ipc_requested()) {
    std::random_device rd;
    const std::string nm = "/skl_" + std::to_string((long long)getpid()) + "_" + std::to_string(rd()) +
                           std::to_string(rd());
    std::memset(out128, 0, 128);
    std::memcpy(out128, nm.c_str(), std::min<size_t>(nm.size(), 127));
    return;
  }
  ncclUniqueId id;
  nccl_check(nccl()->getUniqueId(&id), "ncclGetUniqueId");
  std::memcpy(out128, &id, sizeof(id));
}

void nccl_init(Ctx* ctx, const void* id128) {
  if (!id128) fail(SKL_ERR_INVALID_ARG, "multi-process mode needs the NCCL unique id");
  if (shm_mode()) {
    shm_init(ctx, id128);
    return;
  }
  if (ipc_requested()) {
    ipc_init(ctx, id128);
    return;
  }
  ncclUniqueId id;
  std::memcpy(&id, id128, sizeof(id));
  ctx->set_device(ctx->first_local);
  ncclComm_t comm = nullptr;
  nccl_check(nccl()->commInitRank(&comm, ctx->world, id, ctx->rank), "ncclCommInitRank");
  ctx->nccl_comm = comm;
}

void nccl_destroy(Ctx* ctx) {
  shm_destroy(ctx);
  ipc_destroy(ctx);
  if (ctx->nccl_comm) nccl()->commDestroy((ncclComm_t)ctx->nccl_comm);
  ctx->nccl_comm = nullptr;
}

void run_transfers(Ctx* ctx, const std::vector<Transfer>& tr, size_t unit_bytes, PtrFn& p) {
  if (tr.empty()) return;
  if (!ctx->dist_mode) {
    // one process: the moves into each device run as ONE batched copy kernel on
    // that device's stream (same-GPU sources, or peer loads over NVLink);
    // sources without peer access use the copy engines
    barrier_streams(ctx);
    // one launch per PHYSICAL destination GPU (logical devices sharing a GPU
    // are served by one kernel on the first one's stream; the barriers around
    // order it with every device stream)
    std::vector<int> launcher((size_t)ctx->G);
    for (int g = 0; g < ctx->G; ++g) {
      launcher[(size_t)g] = g;
      for (int h = 0; h < g; ++h)
        if (ctx->D(h).phys == ctx->D(g).phys) {
          launcher[(size_t)g] = h;
          break;
        }
    }
    std::vector<std::vector<XferSeg>> batch((size_t)ctx->G);
    for (const Transfer& t : tr) {
      const size_t bytes = t.n * unit_bytes;
      if (bytes == 0) continue;
      Device& S = ctx->D(t.src);
      Device& D = ctx->D(t.dst);
      void* s = p.src(t);
      void* d = p.dst(t);
      ctx->p2p += (long long)bytes;
      const int lg = launcher[(size_t)t.dst];
      if (ctx->xfer_kernel && ctx->peer_ok[(size_t)lg][(size_t)t.src]) {
        batch[(size_t)lg].push_back(XferSeg{s, d, bytes});
        continue;
      }
      SKL_CUDA(cudaSetDevice(D.phys));
      if (S.phys == D.phys)
        SKL_CUDA(cudaMemcpyAsync(d, s, bytes, cudaMemcpyDeviceToDevice, D.stream));
      else
        SKL_CUDA(cudaMemcpyPeerAsync(d, D.phys, s, S.phys, bytes, D.stream));
    }
    for (int g = 0; g < ctx->G; ++g)
      if (!batch[(size_t)g].empty()) launch_xfer_batch(ctx, g, batch[(size_t)g]);
    barrier_streams(ctx);
    return;
  }
  if (ctx->ipc) {
    // one process per GPU over NVLink peer memory: every rank publishes the
    // addresses of the moves it sources (host exchange, in list order), the
    // device barrier makes every source final on every GPU, then each rank
    // pulls the moves into it with ONE batched copy kernel (peer loads), and a
    // second barrier keeps the sources alive until every rank has read them
    const int me = ctx->first_local;
    std::vector<uint64_t> mine(tr.size(), 0);
    for (size_t i = 0; i < tr.size(); ++i)
      if (tr[i].src == me && tr[i].n) mine[i] = (uint64_t)(uintptr_t)p.src(tr[i]);
    const auto all = ipc_exchange(ctx, mine);
    ipc_barrier(ctx);
    std::vector<XferSeg> segs;
    for (size_t i = 0; i < tr.size(); ++i) {
      const Transfer& t = tr[i];
      const size_t bytes = t.n * unit_bytes;
      if (bytes == 0 || t.dst != me) continue;
      const void* src = t.src == me ? p.src(t) : ipc_translate(ctx, t.src, all[(size_t)t.src].at(i));
      if (t.src != me) ctx->p2p += (long long)bytes;
      segs.push_back(XferSeg{src, p.dst(t), bytes});
    }
    if (!segs.empty()) launch_xfer_batch(ctx, me, segs);
    ipc_barrier(ctx);
    return;
  }
  if (ctx->shm_comm) {
    auto* sc = (ShmComm*)ctx->shm_comm;
    Device& L = ctx->D(ctx->first_local);
    ctx->set_device(ctx->first_local);
    for (const Transfer& t : tr) {
      const size_t bytes = t.n * unit_bytes;
      if (bytes == 0) continue;
      const bool src_here = ctx->is_local(t.src), dst_here = ctx->is_local(t.dst);
      if (src_here && dst_here) {
        SKL_CUDA(cudaMemcpyAsync(p.dst(t), p.src(t), bytes, cudaMemcpyDeviceToDevice, L.stream));
      } else if (src_here) {
        shm_send(ctx, *sc, p.src(t), bytes, t.dst);
        ctx->p2p += (long long)bytes;
      } else if (dst_here) {
        shm_recv(ctx, *sc, p.dst(t), bytes, t.src);
      }
    }
    return;
  }
  NcclApi* a = nccl();
  ncclComm_t comm = (ncclComm_t)ctx->nccl_comm;
  Device& L = ctx->D(ctx->first_local);
  ctx->set_device(ctx->first_local);
  nccl_check(a->groupStart(), "ncclGroupStart");
  for (const Transfer& t : tr) {
    const size_t bytes = t.n * unit_bytes;
    if (bytes == 0) continue;
    const bool src_here = ctx->is_local(t.src), dst_here = ctx->is_local(t.dst);
    if (src_here && dst_here) {
      SKL_CUDA(cudaMemcpyAsync(p.dst(t), p.src(t), bytes,
                               cudaMemcpyDeviceToDevice, L.stream));
    } else if (src_here) {
      nccl_check(a->send(p.src(t), bytes, ncclUint8, t.dst, comm, L.stream), "ncclSend");
      ctx->p2p += (long long)bytes;
    } else if (dst_here) {
      nccl_check(a->recv(p.dst(t), bytes, ncclUint8, t.src, comm, L.stream), "ncclRecv");
    }
  }
  nccl_check(a->groupEnd(), "ncclGroupEnd");
  ctx->n_nccl_group++;
  // errors of communication already in flight (peer failure, transport errors)
  if (a->asyncError) {
    ncclResult_t ar = ncclSuccess;
    nccl_check(a->asyncError(comm, &ar), "ncclCommGetAsyncError");
    if (ar != ncclSuccess && ar != ncclInProgress) nccl_check(ar, "NCCL asynchronous error");
  }
}

}  // namespace skl
