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
#include <nccl.h>

#include <mutex>

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
    const char* names[] = {"libnccl.so.2", "/usr/lib/x86_64-linux-gnu/libnccl.so.2", "libnccl.so"};
    for (const char* n : names) {
      a.h = dlopen(n, RTLD_NOW | RTLD_GLOBAL);
      if (a.h) break;
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

void nccl_get_unique_id(void* out128) {
  ncclUniqueId id;
  nccl_check(nccl()->getUniqueId(&id), "ncclGetUniqueId");
  std::memcpy(out128, &id, sizeof(id));
}

void nccl_init(Ctx* ctx, const void* id128) {
  if (!id128) fail(SKL_ERR_INVALID_ARG, "multi-process mode needs the NCCL unique id");
  ncclUniqueId id;
  std::memcpy(&id, id128, sizeof(id));
  ctx->set_device(ctx->first_local);
  ncclComm_t comm = nullptr;
  nccl_check(nccl()->commInitRank(&comm, ctx->world, id, ctx->rank), "ncclCommInitRank");
  ctx->nccl_comm = comm;
}

void nccl_destroy(Ctx* ctx) {
  if (ctx->nccl_comm) nccl()->commDestroy((ncclComm_t)ctx->nccl_comm);
  ctx->nccl_comm = nullptr;
}

void run_transfers(Ctx* ctx, const std::vector<Transfer>& tr, size_t unit_bytes, PtrFn& p) {
  if (tr.empty()) return;
  if (!ctx->dist_mode) {
    barrier_streams(ctx);
    for (const Transfer& t : tr) {
      const size_t bytes = t.n * unit_bytes;
      if (bytes == 0) continue;
      Device& S = ctx->D(t.src);
      Device& D = ctx->D(t.dst);
      void* s = p.src(t);
      void* d = p.dst(t);
      SKL_CUDA(cudaSetDevice(D.phys));
      if (S.phys == D.phys)
        SKL_CUDA(cudaMemcpyAsync(d, s, bytes, cudaMemcpyDeviceToDevice, D.stream));
      else
        SKL_CUDA(cudaMemcpyPeerAsync(d, D.phys, s, S.phys, bytes, D.stream));
      ctx->p2p += (long long)bytes;
    }
    barrier_streams(ctx);
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
  // errors of communication already in flight (peer failure, transport errors)
  if (a->asyncError) {
    ncclResult_t ar = ncclSuccess;
    nccl_check(a->asyncError(comm, &ar), "ncclCommGetAsyncError");
    if (ar != ncclSuccess && ar != ncclInProgress) nccl_check(ar, "NCCL asynchronous error");
  }
}

}  // namespace skl
