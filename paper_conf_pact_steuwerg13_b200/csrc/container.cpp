// container.cpp — containers, implicit transfers and the redistribution engine
// (SURVEY §1 layers B2/B3).
//
// Vector / Matrix containers; "when a container is created on the
// CPU, memory is allocated on the GPUs automatically".  P:L158-168: transfers
// CPU<->GPU happen implicitly: before a skeleton reads a container and before
// the host reads it.  P:L223-231: a container's distribution can change at run
// time and SkelCL moves the data.  Reading A25: leaving a copy distribution whose
// replicas diverged folds them with the combine function, in GPU order.
//
// Storage model: device g's part is one buffer covering a unit range `buf`
// (units = elements of a vector, rows of a matrix); `valid` is the sub-range
// holding data.  A part may keep spare halo room so that block -> overlap(d)
// (the halo refresh of iterated stencils) moves only the 2d border units.
#include <algorithm>

#include "skl_internal.h"

namespace skl {

void launch_fill(Ctx* ctx, int g, void* dst, size_t bytes, const void* pattern, size_t elt);

Cont* cont_create(Ctx* ctx, int type, size_t rows, size_t cols, bool matrix) {
  const TypeInfo& ti = ctx->type(type);
  if (ti.size == 0) fail(SKL_ERR_TYPE, "containers cannot hold void");
  auto* c = new Cont();
  c->ctx = ctx;
  c->type = type;
  c->elt = ti.size;
  c->matrix = matrix;
  c->rows = rows;
  c->cols = matrix ? cols : 1;
  c->parts.resize((size_t)ctx->G);
  ctx->conts.insert(c);
  return c;
}

// device stream of g waits for the pending chunks of one part
static void sync_part(Cont* c, int g) {
  Part& p = c->parts[(size_t)g];
  if (p.ready.empty()) return;
  Ctx* ctx = c->ctx;
  ctx->set_device(g);
  for (const Ready& rd : p.ready) {
    SKL_CUDA(cudaStreamWaitEvent(ctx->D(g).stream, rd.ev, 0));
    event_put(ctx, g, rd.ev);
  }
  p.ready.clear();
}

void sync_ready(Cont* c) {
  Ctx* ctx = c->ctx;
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g)
    if ((size_t)g < c->parts.size()) sync_part(c, g);
}

// number of chunks for a host<->device transfer of `bytes` (1 = one copy on the
// device stream): chunks let a Map start on the first rows while the rest is in
// flight, and stream its output back while later rows compute
static int xfer_chunks(Ctx* ctx, size_t bytes) {
  if (ctx->capturing || ctx->xfer_chunks <= 1 || bytes < (size_t)(4u << 20)) return 1;
  return (int)std::min<size_t>((size_t)ctx->xfer_chunks, bytes / (1u << 20));
}
// chunk k of K of the unit range r (boundaries on multiples of 64 units, so
// that chunk pointers keep the buffer's 16-byte alignment).  Tapered (default,
// option xfer_taper): the last two chunks are 1/4 and 1/2 of the others, so the
// work that follows the last upload - computing the last chunk and streaming
// its result back - is short (the end-to-end step of a Map whose input and
// output cross PCIe is the upload time plus that tail).
static Range chunk_of(Ctx* ctx, const Range& r, int k, int K) {
  // weights in quarters: 4 for every chunk but the last two (2, 1)
  const bool taper = ctx->xfer_taper && K >= 4;
  const size_t total = taper ? (size_t)4 * (size_t)(K - 2) + 3 : (size_t)K;
  auto cum = [&](int i) -> size_t {  // weight of chunks [0, i)
    if (!taper) return (size_t)i;
    if (i <= K - 2) return (size_t)4 * (size_t)i;
    return (size_t)4 * (size_t)(K - 2) + (i == K - 1 ? 2 : 3);
  };
  auto cut = [&](int i) -> size_t {
    if (i >= K) return r.hi;
    return r.lo + (r.size() * cum(i) / total) / 64 * 64;
  };
  return Range{cut(k), cut(k + 1)};
}

static void free_part(Cont* c, int g) {
  sync_part(c, g);  // pending copies into the buffer complete before it is freed
  Part& p = c->parts[(size_t)g];
  if (p.ptr) device_free(c->ctx, g, p.ptr);
  p = Part();
}

void cont_destroy(Cont* c) {
  Ctx* ctx = c->ctx;
  materialize_dependents(c);
  drop_lazy(c);
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) free_part(c, g);
  for (size_t g = 0; g < c->stage.size(); ++g)
    if (c->stage[g]) device_free(ctx, (int)g, c->stage[g]);
  if (c->host) cudaFreeHost(c->host);
  ctx->conts.erase(c);
  delete c;
}

void* part_ptr(Cont* c, int g, size_t unit) {
  Part& p = c->parts[(size_t)g];
  if (!p.ptr || unit < p.buf.lo || unit > p.buf.hi)
    fail(SKL_ERR_DISTRIBUTION, "internal: unit " + std::to_string(unit) + " not stored on device " +
                                   std::to_string(g));
  return (char*)p.ptr + (unit - p.buf.lo) * c->unit_bytes();
}

static Range alloc_range(Cont* c, const Dist& d, int g) {
  Range need = need_range(c->units(), c->ctx->G, d, g);
  if (need.empty()) return need;
  if ((d.kind == DBLOCK || d.kind == DOVERLAP) && c->spare_halo) {
    const Range core = core_range(c->units(), c->ctx->G, d, g);
    const size_t s = c->spare_halo;
    need.lo = std::min(need.lo, core.lo >= s ? core.lo - s : 0);
    need.hi = std::max(need.hi, std::min(c->units(), core.hi + s));
  }
  return need;
}

// (Re)allocate device parts for layout d; data in reused buffers is kept.
static void set_layout(Cont* c, const Dist& d) {
  Ctx* ctx = c->ctx;
  sync_ready(c);
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) {
    const Range ar = alloc_range(c, d, g);
    Part& p = c->parts[(size_t)g];
    if (ar.empty()) {
      free_part(c, g);
      continue;
    }
    if (p.ptr && p.buf.contains(ar)) continue;
    free_part(c, g);
    p.ptr = device_alloc(ctx, g, ar.size() * c->unit_bytes());
    p.buf = ar;
    p.cap_bytes = ar.size() * c->unit_bytes();
  }
}

static void set_valid(Cont* c, const Dist& d, bool halo) {
  Ctx* ctx = c->ctx;
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) {
    c->parts[(size_t)g].valid =
        halo ? need_range(c->units(), ctx->G, d, g) : core_range(c->units(), ctx->G, d, g);
  }
}

void mark_written(Cont* c) {
  c->dev_valid = true;
  c->host_valid = false;
  c->halo_valid = false;
  c->halo_ready = 0;
  set_valid(c, c->dist, false);
}

void prepare_output(Cont* c, const Dist& d, size_t spare) {
  materialize_dependents(c);  // deferred readers of c's old value run first
  drop_lazy(c);               // a deferred value of c itself is discarded
  if (spare > c->spare_halo) c->spare_halo = spare;
  // buffers that must move would lose data; outputs are overwritten anyway
  set_layout(c, d);
  c->dist = d;
  c->diverged = false;
  c->dev_valid = false;
  c->halo_valid = false;
  c->halo_ready = 0;
}

// ------------------------------------------------------------------ host <-> device
void host_upload(Cont* c, const void* host) {
  Ctx* ctx = c->ctx;
  const size_t ub = c->unit_bytes();
  Dist d = c->dist;
  if (d.kind == DCOPY && ctx->G > 1) {
    // one PCIe upload, then replicate device-to-device over NVLink: upload the
    // block slices (each device its own) and all-gather them.
    Dist b{DBLOCK, 0};
    c->dist = b;
    host_upload(c, host);
    c->diverged = false;
    ensure(c, d, false);
    return;
  }
  set_layout(c, d);
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) {
    const Range r = need_range(c->units(), ctx->G, d, g);
    if (r.empty()) continue;
    ctx->set_device(g);
    Device& D = ctx->D(g);
    const int K = xfer_chunks(ctx, r.size() * ub);
    if (K == 1) {
      SKL_CUDA(cudaMemcpyAsync(part_ptr(c, g, r.lo), (const char*)host + r.lo * ub, r.size() * ub,
                               cudaMemcpyHostToDevice, D.stream));
    } else {
      // chunked upload on the copy stream, after whatever the device stream
      // queued on this buffer (its allocation, earlier readers); each chunk's
      // event lets a consumer start on it while later chunks are in flight
      SKL_CUDA(cudaEventRecord(D.ev, D.stream));
      SKL_CUDA(cudaStreamWaitEvent(D.h2d, D.ev, 0));
      Part& p = c->parts[(size_t)g];
      for (int k = 0; k < K; ++k) {
        const Range q = chunk_of(ctx, r, k, K);
        if (q.empty()) continue;
        SKL_CUDA(cudaMemcpyAsync(part_ptr(c, g, q.lo), (const char*)host + q.lo * ub, q.size() * ub,
                                 cudaMemcpyHostToDevice, D.h2d));
        cudaEvent_t e = event_get(ctx, g);
        SKL_CUDA(cudaEventRecord(e, D.h2d));
        p.ready.push_back(Ready{q, e});
      }
    }
    ctx->h2d += (long long)(r.size() * ub);
  }
  set_valid(c, d, true);
  c->dev_valid = true;
  c->halo_valid = true;
  c->halo_ready = 0;
  c->diverged = false;
}

static void sync_local(Ctx* ctx) {
  if (ctx->capturing) fail(SKL_ERR_INVALID_ARG, "host-visible results are not available while capturing a graph");
  for (auto& d : ctx->dev) {
    SKL_CUDA(cudaSetDevice(d.phys));
    SKL_CUDA(cudaStreamSynchronize(d.stream));
    SKL_CUDA(cudaStreamSynchronize(d.d2h));
  }
}

// Chunked download of units r of part g to `host` (which receives unit r.lo
// first) on the copy stream, each chunk as soon as its producer finished, when
// the part's pending chunks cover r; returns false (nothing done) otherwise.
static bool stream_out(Cont* c, int g, const Range& r, void* host) {
  Ctx* ctx = c->ctx;
  Part& p = c->parts[(size_t)g];
  if (p.ready.empty() || ctx->capturing) return false;
  size_t covered = 0;
  for (const Ready& rd : p.ready) {
    const size_t lo = std::max(rd.r.lo, r.lo), hi = std::min(rd.r.hi, r.hi);
    if (hi > lo) covered += hi - lo;
  }
  if (covered != r.size()) return false;  // chunks overlap or leave gaps: plain path
  ctx->set_device(g);
  Device& D = ctx->D(g);
  const size_t ub = c->unit_bytes();
  for (const Ready& rd : p.ready) {
    const size_t lo = std::max(rd.r.lo, r.lo), hi = std::min(rd.r.hi, r.hi);
    SKL_CUDA(cudaStreamWaitEvent(D.d2h, rd.ev, 0));
    if (hi > lo)
      SKL_CUDA(cudaMemcpyAsync((char*)host + (lo - r.lo) * ub, part_ptr(c, g, lo), (hi - lo) * ub,
                               cudaMemcpyDeviceToHost, D.d2h));
    event_put(ctx, g, rd.ev);
  }
  p.ready.clear();
  // later writers of this buffer on the device stream come after the reads
  SKL_CUDA(cudaEventRecord(D.ev, D.d2h));
  SKL_CUDA(cudaStreamWaitEvent(D.stream, D.ev, 0));
  return true;
}

namespace {
struct ContPtrs : PtrFn {
  Cont* src_c;
  std::vector<Part>* src_parts;  // old parts (may differ from src_c->parts)
  Cont* dst_c;
  void* src(const Transfer& t) override {
    Part& p = (*src_parts)[(size_t)t.src];
    return (char*)p.ptr + (t.src_unit - p.buf.lo) * src_c->unit_bytes();
  }
  void* dst(const Transfer& t) override { return part_ptr(dst_c, t.dst, t.dst_unit); }
};
// gather everything into one full-size buffer on the local device (dist mode)
struct GatherPtrs : PtrFn {
  Cont* c;
  void* buf;
  void* src(const Transfer& t) override { return part_ptr(c, t.src, t.src_unit); }
  void* dst(const Transfer& t) override { return (char*)buf + t.dst_unit * c->unit_bytes(); }
};
}  // namespace

void host_download(Cont* c, void* host) {
  Ctx* ctx = c->ctx;
  if (ctx->capturing) fail(SKL_ERR_INVALID_ARG, "host-visible results are not available while capturing a graph");
  materialize(c);
  const size_t ub = c->unit_bytes();
  if (!c->dev_valid) {
    if (c->host_valid && c->host && host != c->host) std::memcpy(host, c->host, c->bytes());
    else if (!c->host_valid) std::memset(host, 0, c->bytes());
    return;
  }
  if (c->dist.kind == DCOPY && c->diverged && c->combine) copy_combine_to_copy(c);
  if (!ctx->dist_mode) {
    for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) {
      // each unit from its owner (copy: device g's block slice, parallel D2H)
      Range r = c->dist.kind == DCOPY ? block_range(c->units(), ctx->G, g)
                                      : core_range(c->units(), ctx->G, c->dist, g);
      if (r.empty()) continue;
      if (!stream_out(c, g, r, (char*)host + r.lo * ub)) {
        ctx->set_device(g);
        SKL_CUDA(cudaMemcpyAsync((char*)host + r.lo * ub, part_ptr(c, g, r.lo), r.size() * ub,
                                 cudaMemcpyDeviceToHost, ctx->D(g).stream));
      }
      ctx->d2h += (long long)(r.size() * ub);
    }
    sync_local(ctx);
    return;
  }
  sync_ready(c);
  // one process per GPU: every rank assembles the whole container (collective)
  const int g = ctx->first_local;
  const Range have = core_range(c->units(), ctx->G, c->dist, g);
  if (c->dist.kind == DCOPY) {
    ctx->set_device(g);
    SKL_CUDA(cudaMemcpyAsync(host, part_ptr(c, g, 0), c->bytes(), cudaMemcpyDeviceToHost, ctx->D(g).stream));
    ctx->d2h += (long long)c->bytes();
    sync_local(ctx);
    return;
  }
  void* buf = device_alloc(ctx, g, c->bytes());
  if (!have.empty()) {
    ctx->set_device(g);
    SKL_CUDA(cudaMemcpyAsync((char*)buf + have.lo * ub, part_ptr(c, g, have.lo), have.size() * ub,
                             cudaMemcpyDeviceToDevice, ctx->D(g).stream));
  }
  const std::vector<Transfer> tr =
      plan_transfers(c->units(), ctx->G, c->dist, false, Dist{DCOPY, 0}, false);
  GatherPtrs gp;
  gp.c = c;
  gp.buf = buf;
  run_transfers(ctx, tr, ub, gp);
  ctx->set_device(g);
  SKL_CUDA(cudaMemcpyAsync(host, buf, c->bytes(), cudaMemcpyDeviceToHost, ctx->D(g).stream));
  ctx->d2h += (long long)c->bytes();
  device_free(ctx, g, buf);
  sync_local(ctx);
}

void download_part(Cont* c, int g, void* host, size_t* first, size_t* n) {
  Ctx* ctx = c->ctx;
  if (!ctx->is_local(g)) fail(SKL_ERR_INVALID_ARG, "device is not local to this process");
  materialize(c);
  if (!c->dev_valid) fail(SKL_ERR_DISTRIBUTION, "container has no device data");
  if (c->dist.kind == DCOPY && c->diverged && c->combine) copy_combine_to_copy(c);
  const Range r = core_range(c->units(), ctx->G, c->dist, g);
  *first = r.lo;
  *n = r.size();
  if (r.empty()) return;
  ctx->set_device(g);
  if (stream_out(c, g, r, host)) {
    SKL_CUDA(cudaStreamSynchronize(ctx->D(g).d2h));
  } else {
    SKL_CUDA(cudaMemcpyAsync(host, part_ptr(c, g, r.lo), r.size() * c->unit_bytes(),
                             cudaMemcpyDeviceToHost, ctx->D(g).stream));
  }
  ctx->d2h += (long long)(r.size() * c->unit_bytes());
  SKL_CUDA(cudaStreamSynchronize(ctx->D(g).stream));
}

void* host_mirror(Cont* c, int mode) {
  if (mode & SKL_WRITE) materialize_dependents(c);
  if (mode & SKL_READ) materialize(c);
  else drop_lazy(c);
  if (!c->host) SKL_CUDA(cudaHostAlloc(&c->host, std::max<size_t>(c->bytes(), 1), cudaHostAllocPortable));
  if ((mode & SKL_READ) && !c->host_valid) {
    host_download(c, c->host);
    c->host_valid = true;
  }
  if (mode & SKL_WRITE) {
    c->host_valid = true;
    c->dev_valid = false;  // devices become stale
    c->halo_ready = 0;
    c->diverged = false;
  }
  return c->host;
}

void fill(Cont* c, const void* value) {
  Ctx* ctx = c->ctx;
  materialize_dependents(c);
  drop_lazy(c);
  if (c->dist.kind == DNONE) {
    char* h = (char*)host_mirror(c, SKL_WRITE);
    for (size_t i = 0; i < c->rows * c->cols; ++i) std::memcpy(h + i * c->elt, value, c->elt);
    return;
  }
  set_layout(c, c->dist);
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) {
    Part& p = c->parts[(size_t)g];
    if (!p.ptr) continue;
    launch_fill(ctx, g, p.ptr, p.buf.size() * c->unit_bytes(), value, c->elt);
  }
  set_valid(c, c->dist, true);
  c->dev_valid = true;
  c->halo_valid = true;
  c->halo_ready = 0;
  c->host_valid = false;
  c->diverged = false;
}

// ------------------------------------------------------------------ redistribution
// copy(+) -> block (reading A25): block g = r_0[g] (+) ... (+) r_{G-1}[g].
// Every device gathers the G replica slices of its block into staging (one
// canonical all-to-all), then the ordered-combine kernel folds them.
static void combine_to_block(Cont* c) {
  Ctx* ctx = c->ctx;
  sync_ready(c);
  const int G = ctx->G;
  const size_t U = c->units(), ub = c->unit_bytes();
  const Dist blk{DBLOCK, 0};
  if (G == 1) {  // the fold of a single replica is the replica itself
    c->dist = blk;
    c->diverged = false;
    set_valid(c, blk, false);
    return;
  }
  // one process driving every device, each able to load from every replica,
  // <= 8 replicas: one fused exchange + fold kernel per device (peer loads), the
  // fold written in place into the device's own replica
  if (ctx->ipc && ctx->combine_peer && ctx->xfer_kernel) {
    // one process per GPU over NVLink: the same fused exchange + fold, every
    // rank reading the peers' replicas through the IPC mappings
    const int me = ctx->first_local;
    const Part& p = c->parts[(size_t)me];
    const bool ok = p.ptr && p.buf.contains(Range{0, U});
    const auto all = ipc_exchange(ctx, {(uint64_t)(uintptr_t)p.ptr, (uint64_t)p.buf.lo, ok ? 1u : 0u});
    bool all_ok = G <= 8;
    for (int h = 0; h < G; ++h) all_ok = all_ok && all[(size_t)h].at(2) == 1;
    if (all_ok) {
      NvtxRange nr("skl_combine_peer");
      const Range r = block_range(U, G, me);
      ipc_barrier(ctx);  // every replica is final before any rank reads it
      if (!r.empty()) {
        std::vector<const void*> srcs((size_t)G);
        for (int h = 0; h < G; ++h)
          srcs[(size_t)h] = (const char*)ipc_translate(ctx, h, all[(size_t)h][0]) + (r.lo - all[(size_t)h][1]) * ub;
        ctx->p2p += (long long)((size_t)(G - 1) * r.size() * ub);
        run_combine_peer(c->combine, me, srcs.data(), G, part_ptr(c, me, r.lo), r.size() * c->cols);
      }
      ipc_barrier(ctx);  // no rank overwrites its replica while a peer still reads it
      if (r.empty()) free_part(c, me);
      c->dist = blk;
      c->diverged = false;
      c->dev_valid = true;
      c->halo_valid = false;
      c->halo_ready = 0;
      set_valid(c, blk, false);
      return;
    }
  }
  bool fused = ctx->combine_peer && ctx->xfer_kernel && !ctx->dist_mode && ctx->nlocal == G && G <= 8;
  for (int g = 0; fused && g < G; ++g)
    for (int h = 0; h < G; ++h)
      fused = fused && ctx->peer_ok[(size_t)g][(size_t)h] && c->parts[(size_t)h].ptr &&
              c->parts[(size_t)h].buf.contains(Range{0, U});
  if (fused) {
    NvtxRange nr("skl_combine_peer");
    barrier_streams(ctx);  // every replica is final before any device reads it
    std::vector<const void*> srcs((size_t)G);
    bool one_gpu = ctx->combine_peer != 2;  // 2: one kernel per device even on one GPU (tests)
    for (int g = 0; g < G; ++g) one_gpu = one_gpu && ctx->D(g).phys == ctx->D(0).phys;
    if (one_gpu) {
      // logical devices of one GPU: every slice folded by one launch
      for (int h = 0; h < G; ++h) srcs[(size_t)h] = part_ptr(c, h, 0);
      ctx->p2p += (long long)((size_t)(G - 1) * U * ub);
      run_combine_all(c->combine, 0, srcs.data(), G, U * c->cols, (U + (size_t)G - 1) / (size_t)G * c->cols);
    }
    for (int g = 0; g < G && !one_gpu; ++g) {
      const Range r = block_range(U, G, g);
      if (r.empty()) continue;
      for (int h = 0; h < G; ++h) srcs[(size_t)h] = part_ptr(c, h, r.lo);
      ctx->p2p += (long long)((size_t)(G - 1) * r.size() * ub);
      run_combine_peer(c->combine, g, srcs.data(), G, part_ptr(c, g, r.lo), r.size() * c->cols);
    }
    barrier_streams(ctx);  // no device overwrites its replica while a peer still reads it
    for (int g = 0; g < G; ++g)
      if (block_range(U, G, g).empty()) free_part(c, g);
    c->dist = blk;
    c->diverged = false;
    c->dev_valid = true;
    c->halo_valid = false;
    c->halo_ready = 0;
    set_valid(c, blk, false);
    return;
  }
  std::vector<void*> staging((size_t)G, nullptr);
  std::vector<Transfer> tr;
  for (int g = 0; g < G; ++g) {
    const Range r = block_range(U, G, g);
    if (r.empty()) continue;
    for (int h = 0; h < G; ++h) tr.push_back(Transfer{h, g, r.lo, r.lo, r.size(), h});
  }
  // staging slots of device g: G replica slices, each padded to a multiple of
  // 16 elements (so every slot starts 16-byte aligned for the vector combine)
  auto slot_elems = [&](const Range& r) { return (r.size() * c->cols + 15) / 16 * 16; };
  // staging is kept with the container between combines (LM OSEM combines
  // every subset): no allocation on the steady-state path
  c->stage.resize((size_t)G, nullptr);
  c->stage_bytes.resize((size_t)G, 0);
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) {
    const Range r = block_range(U, G, g);
    if (r.empty()) continue;
    const size_t need = (size_t)G * slot_elems(r) * c->elt;
    if (c->stage_bytes[(size_t)g] < need) {
      device_free(ctx, g, c->stage[(size_t)g]);
      c->stage[(size_t)g] = device_alloc(ctx, g, need);
      c->stage_bytes[(size_t)g] = need;
    }
    staging[(size_t)g] = c->stage[(size_t)g];
  }
  struct StagePtrs : PtrFn {
    Cont* c;
    std::vector<void*>* st;
    size_t U;
    int G;
    void* src(const Transfer& t) override { return part_ptr(c, t.src, t.src_unit); }
    void* dst(const Transfer& t) override {
      const Range r = block_range(U, G, t.dst);
      const size_t slot = (r.size() * c->cols + 15) / 16 * 16 * c->elt;
      return (char*)(*st)[(size_t)t.dst] + (size_t)t.slot * slot + (t.dst_unit - r.lo) * c->unit_bytes();
    }
  } sp;
  sp.c = c;
  sp.st = &staging;
  sp.U = U;
  sp.G = G;
  run_transfers(ctx, tr, ub, sp);
  // the folded block of device g goes into its replica's buffer (it covers
  // the block range; every read of that slice went to staging, and the
  // transfers finished at run_transfers' closing barrier)
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) {
    const Range r = block_range(U, G, g);
    const Range ar = alloc_range(c, blk, g);
    Part& p = c->parts[(size_t)g];
    if (r.empty()) {
      free_part(c, g);
      continue;
    }
    if (!p.ptr || !p.buf.contains(ar)) {
      free_part(c, g);
      p.ptr = device_alloc(ctx, g, ar.size() * ub);
      p.buf = ar;
      p.cap_bytes = ar.size() * ub;
    }
    run_combine(c->combine, g, staging[(size_t)g], slot_elems(r), G, part_ptr(c, g, r.lo), r.size() * c->cols);
  }
  c->dist = blk;
  c->diverged = false;
  c->dev_valid = true;
  c->halo_valid = false;
  c->halo_ready = 0;
  set_valid(c, blk, false);
}

static void redistribute(Cont* c, const Dist& to) {
  NvtxRange nr("skl_redistribute");
  Ctx* ctx = c->ctx;
  const size_t U = c->units(), ub = c->unit_bytes();
  const Dist from = c->dist;
  const bool from_halo = from.kind == DOVERLAP && c->halo_valid;
  const bool to_halo = to.kind == DOVERLAP;
  const std::vector<Transfer> tr = plan_transfers(U, ctx->G, from, from_halo, to, to_halo);
  std::vector<Part> old = c->parts;
  std::vector<bool> moved((size_t)ctx->G, false);
  // new layout; keep buffers that already cover the target
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) {
    const Range ar = alloc_range(c, to, g);
    Part& p = c->parts[(size_t)g];
    if (ar.empty()) {
      if (p.ptr) moved[(size_t)g] = true;  // freed after the exchange
      p = Part();
      continue;
    }
    if (p.ptr && p.buf.contains(ar)) continue;
    moved[(size_t)g] = p.ptr != nullptr;
    p = Part();
    p.ptr = device_alloc(ctx, g, ar.size() * ub);
    p.buf = ar;
    p.cap_bytes = ar.size() * ub;
    // units this device already holds move locally into the new buffer
    const Range have = from_halo ? need_range(U, ctx->G, from, g) : core_range(U, ctx->G, from, g);
    const Range want = to_halo ? need_range(U, ctx->G, to, g) : core_range(U, ctx->G, to, g);
    const Range keep{std::max(have.lo, want.lo), std::min(have.hi, want.hi)};
    const Part& o = old[(size_t)g];
    if (!keep.empty() && o.ptr) {
      ctx->set_device(g);
      SKL_CUDA(cudaMemcpyAsync((char*)p.ptr + (keep.lo - p.buf.lo) * ub,
                               (const char*)o.ptr + (keep.lo - o.buf.lo) * ub, keep.size() * ub,
                               cudaMemcpyDeviceToDevice, ctx->D(g).stream));
    }
  }
  ContPtrs cp;
  cp.src_c = c;
  cp.src_parts = &old;
  cp.dst_c = c;
  run_transfers(ctx, tr, ub, cp);
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g)
    if (moved[(size_t)g] && old[(size_t)g].ptr) device_free(ctx, g, old[(size_t)g].ptr);
  c->dist = to;
  c->dev_valid = true;
  c->halo_valid = to_halo;
  c->halo_ready = 0;
  set_valid(c, to, to_halo);
}

static bool halos_allocated(Cont* c, const Dist& d) {
  for (int g = c->ctx->first_local; g < c->ctx->first_local + c->ctx->nlocal; ++g) {
    const Range n = need_range(c->units(), c->ctx->G, d, g);
    const Part& p = c->parts[(size_t)g];
    if (!n.empty() && (!p.ptr || !p.buf.contains(n))) return false;
  }
  return true;
}

static void ensure_impl(Cont* c, const Dist& d, bool halo);

void ensure(Cont* c, const Dist& d, bool halo, bool keep_ready) {
  // nothing to move: pending upload chunks may stay pending for the caller
  const bool noop = !c->lazy.s && c->dev_valid && c->dist == d &&
                    !(d.kind == DOVERLAP && halo && !c->halo_valid) &&
                    !(c->dist.kind == DCOPY && c->diverged && c->combine);
  if (!noop) sync_ready(c);
  ensure_impl(c, d, halo);
  if (!keep_ready) sync_ready(c);
}

static void ensure_impl(Cont* c, const Dist& d, bool halo) {
  if (d.kind == DNONE) fail(SKL_ERR_DISTRIBUTION, "no distribution");
  materialize(c);  // a deferred Zip/Map result is computed before it is used
  if (c->dev_valid && c->dist.kind == DCOPY && c->diverged && c->combine && !(d == c->dist)) {
    combine_to_block(c);
  }
  if (c->dev_valid && c->dist.kind == DCOPY && c->diverged && d.kind == DCOPY && c->combine) {
    copy_combine_to_copy(c);
    return;
  }
  if (c->dev_valid && c->halo_ready && c->dist.kind == DBLOCK && d.kind == DOVERLAP &&
      (size_t)d.arg <= c->halo_ready && halos_allocated(c, d)) {
    // the producing MapOverlap already stored the border units into the
    // neighbours' halo rows (fused halo push): block -> overlap moves nothing
    c->dist = d;
    c->halo_valid = true;
    set_valid(c, d, true);
    return;
  }
  if (c->dist == d && c->dev_valid) {
    if (d.kind == DOVERLAP && halo && !c->halo_valid) {
      // halo refresh: only the border units move
      NvtxRange nr("skl_halo_refresh");
      const std::vector<Transfer> tr = plan_transfers(c->units(), c->ctx->G, d, false, d, true);
      set_layout(c, d);  // buffers already cover the halo (need_range)
      std::vector<Part> cur = c->parts;
      ContPtrs cp;
      cp.src_c = c;
      cp.src_parts = &cur;
      cp.dst_c = c;
      run_transfers(c->ctx, tr, c->unit_bytes(), cp);
      c->halo_valid = true;
      set_valid(c, d, true);
    }
    return;
  }
  if (!c->dev_valid) {
    c->dist = d;
    if (c->host_valid && c->host) {
      host_upload(c, c->host);
    } else {
      // never written: allocate only (contents undefined, A-none)
      set_layout(c, d);
      set_valid(c, d, true);
      c->dev_valid = true;
      c->halo_valid = true;
      c->halo_ready = 0;
    }
    return;
  }
  if (c->dist.kind == DCOPY && c->diverged && !c->combine) c->diverged = false;  // A26
  redistribute(c, d);
}

void copy_combine_to_copy(Cont* c) {
  combine_to_block(c);
  redistribute(c, Dist{DCOPY, 0});
}

}  // namespace skl
