// ipc.cpp — one process per GPU, the data path over NVLink peer memory
// (SKL_COMM=ipc).
//
// In the one-process-per-GPU mode (skl_init_dist) every exchange of the hot path
// - redistribution moves, overlap halo refresh, the
// copy(+) -> block fold (A25), Reduce partials and Scan carries - runs as the
// same in-kernel peer loads / stores the single-process mode uses, instead of
// NCCL send/recv:
//   * device memory of a rank comes from an IPC heap: cudaMalloc'd segments
//     exported once with cudaIpcGetMemHandle and sub-allocated here (first fit,
//     coalescing frees); a peer maps a segment the first time it needs an
//     address inside it (cudaIpcOpenMemHandle) and keeps the mapping;
//   * the ranks of one node share a POSIX shared-memory control block (named by
//     the 128-byte id rank 0 created): per rank the published segment table, a
//     host barrier counter and a double-buffered mailbox through which the
//     ranks exchange device addresses (host barrier, no device work);
//   * a device barrier kernel (one tiny launch on the rank's stream) orders the
//     ranks' streams: each rank stores the barrier epoch into every peer's
//     signal slot (st.release.sys over NVLink) and spins on its own slots
//     (ld.acquire.sys) - the producers of a collective's inputs are complete on
//     every GPU before any rank reads them, and every read is complete before a
//     rank reuses the memory.  A spin gives up after 60 s and raises a sticky
//     host-visible error (SKL_ERR_NCCL at the next collective) instead of
//     hanging the GPU.
// Several ranks may share one GPU (processes time-slice it): the tests run 2-3
// ranks on one B200.
#include <fcntl.h>
#include <sys/mman.h>
#include <unistd.h>

#include <atomic>
#include <chrono>
#include <cstdlib>
#include <thread>

#include "skl_internal.h"

namespace skl {

void launch_ipc_barrier(Ctx* ctx, unsigned long long* const* peer_slots, int world, int rank,
                        unsigned long long* mine, unsigned long long epoch, unsigned* err);  // builtin.cu

namespace {
constexpr int kMaxSegs = 64;
constexpr int kMail = 4096;  // 8-byte words per mailbox

struct ShmSeg {
  unsigned char handle[64];
  uint64_t base, size;
};
struct alignas(64) ShmRank {
  std::atomic<uint64_t> nseg;
  ShmSeg seg[kMaxSegs];
  alignas(64) std::atomic<uint64_t> epoch;  // host barrier arrivals
  alignas(64) uint64_t mail[2][kMail];
};
static_assert(sizeof(cudaIpcMemHandle_t) == 64, "IPC handle size");

struct Seg {
  char* base = nullptr;
  size_t size = 0;
  std::map<size_t, size_t> free;  // offset -> bytes
};
struct PeerSeg {
  uint64_t rbase = 0, size = 0;
  char* local = nullptr;
};

struct Ipc {
  std::string name;
  int rank = 0, world = 1;
  ShmRank* ctl = nullptr;
  size_t ctl_bytes = 0;
  std::vector<Seg> segs;
  std::map<char*, std::pair<int, size_t>> live;  // allocation -> (segment, bytes)
  std::vector<std::vector<PeerSeg>> peers;
  uint64_t host_epoch = 0, dev_epoch = 0;
  unsigned long long* sig = nullptr;                 // my signal slots [kIpcMaxRanks]
  unsigned long long* peer_sig[kIpcMaxRanks] = {};   // each peer's slots, mapped here
  unsigned* err_host = nullptr;                      // pinned, mapped: barrier time-outs
  unsigned* err_dev = nullptr;
};

Ipc& I(Ctx* ctx) {
  if (!ctx->ipc) fail(SKL_ERR_INVALID_ARG, "internal: no IPC transport");
  return *(Ipc*)ctx->ipc;
}

size_t seg_default() {
  if (const char* v = std::getenv("SKL_IPC_SEG_MB")) {
    const long mb = std::strtol(v, nullptr, 10);
    if (mb >= 2 && mb <= (1l << 20)) return (size_t)mb << 20;
  }
  return (size_t)512 << 20;
}

void host_barrier(Ipc& c) {
  const uint64_t e = ++c.host_epoch;
  c.ctl[c.rank].epoch.store(e, std::memory_order_release);
  const auto t0 = std::chrono::steady_clock::now();
  for (int h = 0; h < c.world; ++h) {
    unsigned spins = 0;
    while (c.ctl[h].epoch.load(std::memory_order_acquire) < e) {
      if (++spins > 64) std::this_thread::yield();
      if ((spins & 1023u) == 0 && std::chrono::steady_clock::now() - t0 > std::chrono::seconds(300))
        fail(SKL_ERR_NCCL, "IPC transport: timed out at a host barrier waiting for rank " + std::to_string(h));
    }
  }
}

void new_segment(Ctx* ctx, Ipc& c, size_t bytes) {
  if ((int)c.segs.size() >= kMaxSegs) fail(SKL_ERR_OOM, "IPC heap: segment table full");
  Seg s;
  s.size = std::max(seg_default(), (bytes + (2u << 20) - 1) / (2u << 20) * (2u << 20));
  ctx->set_device(ctx->first_local);
  void* p = nullptr;
  SKL_CUDA(cudaMalloc(&p, s.size));
  s.base = (char*)p;
  s.free[0] = s.size;
  cudaIpcMemHandle_t h;
  SKL_CUDA(cudaIpcGetMemHandle(&h, p));
  const uint64_t k = c.segs.size();
  ShmSeg& out = c.ctl[c.rank].seg[k];
  std::memcpy(out.handle, &h, 64);
  out.base = (uint64_t)(uintptr_t)p;
  out.size = s.size;
  c.ctl[c.rank].nseg.store(k + 1, std::memory_order_release);
  c.segs.push_back(std::move(s));
}
}  // namespace

// The one-process-per-GPU transport: SKL_COMM=ipc (the default: the ranks of
// one node, NVLink peer memory), shm (host loopback, tests) or nccl (NCCL
// send/recv of the same transfer lists, e.g. across nodes).
bool ipc_requested() {
  const char* v = std::getenv("SKL_COMM");
  return !v || !*v || std::string(v) == "ipc";
}

void* ipc_alloc(Ctx* ctx, size_t bytes) {
  Ipc& c = I(ctx);
  bytes = (std::max<size_t>(bytes, 1) + 255) / 256 * 256;
  for (int pass = 0; pass < 2; ++pass) {
    for (size_t si = 0; si < c.segs.size(); ++si) {
      Seg& s = c.segs[si];
      for (auto it = s.free.begin(); it != s.free.end(); ++it) {
        if (it->second < bytes) continue;
        const size_t off = it->first, rest = it->second - bytes;
        s.free.erase(it);
        if (rest) s.free[off + bytes] = rest;
        char* p = s.base + off;
        c.live[p] = {(int)si, bytes};
        return p;
      }
    }
    if (pass == 0) new_segment(ctx, c, bytes);
  }
  fail(SKL_ERR_OOM, "IPC heap: allocation failed");
}

void ipc_free(Ctx* ctx, void* ptr) {
  Ipc& c = I(ctx);
  auto it = c.live.find((char*)ptr);
  if (it == c.live.end()) fail(SKL_ERR_INVALID_ARG, "IPC heap: free of an unknown pointer");
  Seg& s = c.segs[(size_t)it->second.first];
  size_t off = (size_t)((char*)ptr - s.base), len = it->second.second;
  c.live.erase(it);
  // coalesce with the free neighbours
  auto nx = s.free.lower_bound(off);
  if (nx != s.free.end() && nx->first == off + len) {
    len += nx->second;
    nx = s.free.erase(nx);
  }
  if (nx != s.free.begin()) {
    auto pv = std::prev(nx);
    if (pv->first + pv->second == off) {
      pv->second += len;
      return;
    }
  }
  s.free[off] = len;
}

void* ipc_translate(Ctx* ctx, int h, uint64_t va) {
  Ipc& c = I(ctx);
  if (h == c.rank || va == 0) return (void*)(uintptr_t)va;
  for (int pass = 0; pass < 2; ++pass) {
    for (const PeerSeg& s : c.peers[(size_t)h])
      if (va >= s.rbase && va < s.rbase + s.size) return s.local + (va - s.rbase);
    if (pass == 1) break;
    // map the segments rank h published since the last look
    const uint64_t n = c.ctl[h].nseg.load(std::memory_order_acquire);
    ctx->set_device(ctx->first_local);
    for (size_t k = c.peers[(size_t)h].size(); k < n; ++k) {
      const ShmSeg& ss = c.ctl[h].seg[k];
      cudaIpcMemHandle_t hd;
      std::memcpy(&hd, ss.handle, 64);
      void* local = nullptr;
      SKL_CUDA(cudaIpcOpenMemHandle(&local, hd, cudaIpcMemLazyEnablePeerAccess));
      c.peers[(size_t)h].push_back(PeerSeg{ss.base, ss.size, (char*)local});
    }
  }
  fail(SKL_ERR_INVALID_ARG, "IPC transport: address of rank " + std::to_string(h) + " outside its heap");
}

std::vector<std::vector<uint64_t>> ipc_exchange(Ctx* ctx, const std::vector<uint64_t>& mine) {
  Ipc& c = I(ctx);
  if (mine.size() + 1 > (size_t)kMail) fail(SKL_ERR_INVALID_ARG, "IPC transport: exchange too large");
  const int slot = (int)((c.host_epoch + 1) & 1);
  uint64_t* box = c.ctl[c.rank].mail[slot];
  box[0] = mine.size();
  if (!mine.empty()) std::memcpy(box + 1, mine.data(), mine.size() * 8);
  host_barrier(c);  // publishes the mailbox (release) and waits for every rank's
  std::vector<std::vector<uint64_t>> all((size_t)c.world);
  for (int h = 0; h < c.world; ++h) {
    const uint64_t* b = c.ctl[h].mail[slot];
    const size_t n = (size_t)std::min<uint64_t>(b[0], kMail - 1);
    all[(size_t)h].assign(b + 1, b + 1 + n);
  }
  return all;
}

void ipc_check(Ctx* ctx) {
  Ipc& c = I(ctx);
  if (*(volatile unsigned*)c.err_host)
    fail(SKL_ERR_NCCL, "IPC transport: a device barrier timed out (a peer rank stopped participating)");
}

void ipc_barrier(Ctx* ctx) {
  Ipc& c = I(ctx);
  ipc_check(ctx);
  ctx->set_device(ctx->first_local);
  launch_ipc_barrier(ctx, c.peer_sig, c.world, c.rank, c.sig, ++c.dev_epoch, c.err_dev);
}

void ipc_init(Ctx* ctx, const void* id128) {
  if (ctx->world > kIpcMaxRanks) fail(SKL_ERR_UNSUPPORTED, "IPC transport: at most 8 ranks (one node)");
  auto* c = new Ipc();
  ctx->ipc = c;
  c->name = std::string((const char*)id128, strnlen((const char*)id128, 127)) + "_ipc";
  c->rank = ctx->rank;
  c->world = ctx->world;
  c->peers.resize((size_t)c->world);
  c->ctl_bytes = sizeof(ShmRank) * (size_t)c->world;
  const int fd = shm_open(c->name.c_str(), O_CREAT | O_RDWR, 0600);
  if (fd < 0) fail(SKL_ERR_NCCL, "IPC transport: cannot open " + c->name);
  if (ftruncate(fd, (off_t)c->ctl_bytes) != 0) {
    close(fd);
    fail(SKL_ERR_NCCL, "IPC transport: ftruncate failed");
  }
  void* h = mmap(nullptr, c->ctl_bytes, PROT_READ | PROT_WRITE, MAP_SHARED, fd, 0);
  close(fd);
  if (h == MAP_FAILED) fail(SKL_ERR_NCCL, "IPC transport: mmap failed");
  c->ctl = (ShmRank*)h;
  ctx->set_device(ctx->first_local);
  SKL_CUDA(cudaHostAlloc((void**)&c->err_host, sizeof(unsigned), cudaHostAllocMapped));
  *c->err_host = 0u;
  SKL_CUDA(cudaHostGetDevicePointer((void**)&c->err_dev, c->err_host, 0));
  c->sig = (unsigned long long*)ipc_alloc(ctx, kIpcMaxRanks * sizeof(unsigned long long));
  SKL_CUDA(cudaMemset(c->sig, 0, kIpcMaxRanks * sizeof(unsigned long long)));
  SKL_CUDA(cudaDeviceSynchronize());
  const auto all = ipc_exchange(ctx, {(uint64_t)(uintptr_t)c->sig});
  for (int r = 0; r < c->world; ++r)
    c->peer_sig[r] = (unsigned long long*)ipc_translate(ctx, r, all[(size_t)r].at(0));
  ipc_barrier(ctx);  // every rank reaches every other rank's memory
  SKL_CUDA(cudaStreamSynchronize(ctx->D(ctx->first_local).stream));
  ipc_check(ctx);
}

void ipc_destroy(Ctx* ctx) {
  if (!ctx->ipc) return;
  auto* c = (Ipc*)ctx->ipc;
  ctx->set_device(ctx->first_local);
  cudaDeviceSynchronize();
  try {
    host_barrier(*c);  // nobody reads a peer's memory any more
  } catch (const Error&) {
  }
  for (auto& ps : c->peers)
    for (PeerSeg& s : ps) cudaIpcCloseMemHandle(s.local);
  try {
    host_barrier(*c);  // every mapping of my segments is closed
  } catch (const Error&) {
  }
  for (Seg& s : c->segs) cudaFree(s.base);
  if (c->err_host) cudaFreeHost(c->err_host);
  munmap((void*)c->ctl, c->ctl_bytes);
  if (c->rank == 0) shm_unlink(c->name.c_str());
  (void)cudaGetLastError();
  delete c;
  ctx->ipc = nullptr;
}

}  // namespace skl
