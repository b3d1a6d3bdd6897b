// capi.cpp — the C ABI (include/skl.h).  Argument checking and error mapping
// only: every call converts exceptions to skl_status + skl_last_error().
#include <functional>

#include "skl_internal.h"

namespace skl {
Ctx* ctx_create_local(int ndev, const int* devices);
Ctx* ctx_create_dist(int rank, int world, int cuda_device, const void* nccl_id);
Ctx* ctx_create_offline();
void ctx_destroy(Ctx* c);
const char* last_error_cstr();
void set_last_error(const std::string& s);
}  // namespace skl

using namespace skl;


namespace {
template <class F>
skl_status guard(F&& f) {
  try {
    f();
    return SKL_OK;
  } catch (const Error& e) {
    set_last_error(e.what());
    return e.code;
  } catch (const std::bad_alloc&) {
    set_last_error("host allocation failed");
    return SKL_ERR_OOM;
  } catch (const std::exception& e) {
    set_last_error(e.what());
    return SKL_ERR_INVALID_ARG;
  }
}
// Handles map 1:1 onto internal objects; the wrapper structs are owned by them.
std::map<Ctx*, skl_ctx*> g_ctx;
std::map<Cont*, skl_cont*> g_cont;
std::map<Skel*, skl_skel*> g_skel;

Ctx* C(skl_ctx* x) {
  if (!x || !x->c) fail(SKL_ERR_INVALID_ARG, "NULL context");
  return x->c;
}
Cont* K(skl_cont* x) {
  if (!x || !x->c) fail(SKL_ERR_INVALID_ARG, "NULL container");
  return x->c;
}
Skel* S(skl_skel* x) {
  if (!x || !x->s) fail(SKL_ERR_INVALID_ARG, "NULL skeleton");
  return x->s;
}
skl_cont* wrap(Cont* c) {
  auto it = g_cont.find(c);
  if (it != g_cont.end()) return it->second;
  auto* w = new skl_cont{c};
  g_cont[c] = w;
  return w;
}
skl_skel* wrap(Skel* s) {
  auto* w = new skl_skel{s};
  g_skel[s] = w;
  return w;
}
void forget_ctx_objects(Ctx* c) {
  for (auto it = g_cont.begin(); it != g_cont.end();)
    if (it->first->ctx == c) { it->second->c = nullptr; it = g_cont.erase(it); } else ++it;
  for (auto it = g_skel.begin(); it != g_skel.end();)
    if (it->first->ctx == c) { it->second->s = nullptr; it = g_skel.erase(it); } else ++it;
}
// output container handles: NULL -> new container
skl_status run_out(skl_cont** out, const std::function<void(Cont**)>& f) {
  return guard([&] {
    if (!out) fail(SKL_ERR_INVALID_ARG, "NULL output handle pointer");
    Cont* o = *out ? K(*out) : nullptr;
    f(&o);
    *out = wrap(o);
  });
}
}  // namespace

extern "C" {

const char* skl_last_error(void) { return last_error_cstr(); }

skl_status skl_init(int ndev, const int* devices, skl_ctx** out) {
  return guard([&] {
    if (!out) fail(SKL_ERR_INVALID_ARG, "NULL out");
    Ctx* c = ctx_create_local(ndev, devices);
    *out = new skl_ctx{c};
    g_ctx[c] = *out;
  });
}
skl_status skl_init_dist(int rank, int world, int cuda_device, const void* nccl_id, skl_ctx** out) {
  return guard([&] {
    if (!out) fail(SKL_ERR_INVALID_ARG, "NULL out");
    Ctx* c = ctx_create_dist(rank, world, cuda_device, nccl_id);
    *out = new skl_ctx{c};
    g_ctx[c] = *out;
  });
}
skl_status skl_nccl_unique_id(void* out128) {
  return guard([&] {
    if (!out128) fail(SKL_ERR_INVALID_ARG, "NULL out");
    nccl_get_unique_id(out128);
  });
}
skl_status skl_finalize(skl_ctx* ctx) {
  return guard([&] {
    Ctx* c = C(ctx);
    forget_ctx_objects(c);
    ctx_destroy(c);
    g_ctx.erase(c);
    ctx->c = nullptr;
    delete ctx;
  });
}
skl_status skl_num_devices(skl_ctx* ctx, int* ndev, int* first_local, int* nlocal) {
  return guard([&] {
    Ctx* c = C(ctx);
    if (ndev) *ndev = c->G;
    if (first_local) *first_local = c->first_local;
    if (nlocal) *nlocal = c->nlocal;
  });
}
skl_status skl_set_stream(skl_ctx* ctx, int g, void* stream) {
  return guard([&] {
    Ctx* c = C(ctx);
    if (!c->is_local(g)) fail(SKL_ERR_INVALID_ARG, "device is not local");
    Device& d = c->D(g);
    cudaStream_t ns = stream ? (cudaStream_t)stream : d.own;
    if (ns == d.stream) return;
    // order the new stream after everything queued on the old one
    c->set_device(g);
    SKL_CUDA(cudaEventRecord(d.ev, d.stream));
    SKL_CUDA(cudaStreamWaitEvent(ns, d.ev, 0));
    d.stream = ns;
  });
}
skl_status skl_set_allocator(skl_ctx* ctx, skl_alloc_fn alloc, skl_free_fn release, void* user) {
  return guard([&] {
    Ctx* c = C(ctx);
    if ((alloc == nullptr) != (release == nullptr)) fail(SKL_ERR_INVALID_ARG, "give both functions or neither");
    if (!c->conts.empty() || !c->skels.empty())
      fail(SKL_ERR_INVALID_ARG, "set the allocator before creating containers or skeletons");
    c->user_alloc = alloc;
    c->user_free = release;
    c->alloc_user = user;
  });
}
skl_status skl_get_stream(skl_ctx* ctx, int g, void** stream) {
  return guard([&] {
    Ctx* c = C(ctx);
    if (!c->is_local(g) || !stream) fail(SKL_ERR_INVALID_ARG, "bad device or NULL out");
    *stream = (void*)c->D(g).stream;
  });
}
skl_status skl_sync(skl_ctx* ctx) {
  return guard([&] {
    Ctx* c = C(ctx);
    if (c->capturing) fail(SKL_ERR_INVALID_ARG, "skl_sync while capturing a graph");
    for (auto& d : c->dev) {
      SKL_CUDA(cudaSetDevice(d.phys));
      SKL_CUDA(cudaStreamSynchronize(d.stream));
    }
    SKL_CUDA(cudaGetLastError());
  });
}
skl_status skl_set_option(skl_ctx* ctx, const char* key, long long value) {
  return guard([&] {
    Ctx* c = C(ctx);
    const std::string k = key ? key : "";
    if (k == "block_threads") {
      if (value < 64 || value > 1024 || value % 32) fail(SKL_ERR_INVALID_ARG, "block_threads must be a multiple of 32 in [64,1024]");
      c->block_threads = (int)value;
    } else if (k == "debug_bounds") {
      c->debug_bounds = value ? 1 : 0;
    } else if (k == "scan_chunks") {
      if (value != 2 && value != 4 && value != 6 && value != 8 && value != 12 && value != 16)
        fail(SKL_ERR_INVALID_ARG, "scan_chunks in {2,4,6,8,12,16}");
      c->scan_chunks = (int)value;
    } else if (k == "scan_sub") {
      if (value < 1 || value > 64) fail(SKL_ERR_INVALID_ARG, "scan_sub in [1,64]");
      c->scan_sub = (int)value;
    } else if (k == "scan_fstride") {
      if (value < 1 || value > 64) fail(SKL_ERR_INVALID_ARG, "scan_fstride in [1,64]");
      c->scan_fstride = (int)value;
    } else if (k == "scan_spin_ns") {
      if (value < 0 || value > 100000) fail(SKL_ERR_INVALID_ARG, "scan_spin_ns in [0,100000]");
      c->scan_spin_ns = (int)value;
    } else if (k == "scan_lbw") {
      if (value < 1 || value > 8) fail(SKL_ERR_INVALID_ARG, "scan_lbw in [1,8]");
      c->scan_lbw = (int)value;
    } else if (k == "scan_minb_pipe") {
      if (value < 1 || value > 8) fail(SKL_ERR_INVALID_ARG, "scan_minb_pipe in [1,8]");
      c->scan_minb_pipe = (int)value;
    } else if (k == "scan_minb") {
      if (value < 1 || value > 32) fail(SKL_ERR_INVALID_ARG, "scan_minb in [1,32]");
      c->scan_minb = (int)value;
    } else if (k == "mo_persist") {
      c->mo_persist = value ? 1 : 0;
    } else if (k == "mo_ws") {
      c->mo_ws = value ? 1 : 0;
    } else if (k == "map_auto") {
      c->map_auto = value ? 1 : 0;
    } else if (k == "map_il_elems") {
      if (value < 0 || value > 64) fail(SKL_ERR_INVALID_ARG, "map_il_elems in [0,64]");
      c->map_il_elems = (int)value;
    } else if (k == "mo_tma") {
      c->mo_tma = value ? 1 : 0;
    } else if (k == "mo_kt") {
      if (value < 0 || value > 4) fail(SKL_ERR_INVALID_ARG, "mo_kt in [0,4]");
      c->mo_kt = (int)value;
    } else if (k == "mo_full") {
      if (value < -1 || value > 1) fail(SKL_ERR_INVALID_ARG, "mo_full in {-1,0,1}");
      c->mo_full = (int)value;
    } else if (k == "mo_ws_stages") {
      if (value < 2 || value > 8) fail(SKL_ERR_INVALID_ARG, "mo_ws_stages in [2,8]");
      c->mo_ws_stages = (int)value;
    } else if (k == "mo_ws_minb") {
      if (value < 0 || value > 32) fail(SKL_ERR_INVALID_ARG, "mo_ws_minb in [0,32]");
      c->mo_ws_minb = (int)value;
    } else if (k == "mo_minb") {
      if (value < 0 || value > 32) fail(SKL_ERR_INVALID_ARG, "mo_minb in [0,32]");
      c->mo_minb = (int)value;
    } else if (k == "mo_rh" || k == "mo_cw") {
      if (value < 0 || value > 32) fail(SKL_ERR_INVALID_ARG, k + " in [0,32]");
      (k == "mo_rh" ? c->mo_rh : c->mo_cw) = (int)value;
    } else if (k == "lazy_fusion") {
      c->lazy_fusion = value ? 1 : 0;
    } else if (k == "combine_unroll") {
      if (value < 0 || value > 8) fail(SKL_ERR_INVALID_ARG, "combine_unroll in [0,8]");
      c->combine_unroll = (int)value;
    } else if (k == "combine_peer") {
      if (value < 0 || value > 2) fail(SKL_ERR_INVALID_ARG, "combine_peer in {0,1,2}");
      c->combine_peer = (int)value;
    } else if (k == "xfer_kernel") {
      c->xfer_kernel = value ? 1 : 0;
    } else if (k == "xfer_taper") {
      c->xfer_taper = value ? 1 : 0;
    } else if (k == "xfer_chunks") {
      if (value < 1 || value > 64) fail(SKL_ERR_INVALID_ARG, "xfer_chunks in [1,64]");
      c->xfer_chunks = (int)value;
    } else if (k == "map_interleave") {
      c->map_interleave = value ? 1 : 0;
    } else if (k == "ap_bk") {
      if (value != 0 && value != 16 && value != 32) fail(SKL_ERR_INVALID_ARG, "ap_bk in {0,16,32}");
      c->ap_bk = (int)value;
    } else if (k == "ap_hybrid") {
      c->ap_hybrid = value ? 1 : 0;
    } else if (k == "ap_tile") {
      if (value != 0 && value != 2 && value != 4 && value != 8) fail(SKL_ERR_INVALID_ARG, "ap_tile in {0,2,4,8}");
      c->ap_tile = (int)value;
    } else if (k == "ap_fast") {
      c->ap_fast = value ? 1 : 0;
    } else if (k == "halo_push") {
      c->halo_push = value ? 1 : 0;
    } else if (k == "scan_variant") {
      c->scan_variant = (int)value;
    } else if (k == "scan_persistent") {
      c->scan_persistent = value ? 1 : 0;
    } else if (k == "map_unroll") {
      if (value < 1 || value > 16) fail(SKL_ERR_INVALID_ARG, "map_unroll in [1,16]");
      c->map_unroll = (int)value;
    } else {
      fail(SKL_ERR_INVALID_ARG, "unknown option " + k);
    }
  });
}
skl_status skl_get_counter(skl_ctx* ctx, const char* key, long long* value) {
  return guard([&] {
    Ctx* c = C(ctx);
    const std::string k = key ? key : "";
    if (!value) fail(SKL_ERR_INVALID_ARG, "NULL out");
    if (k == "launches") *value = c->n_launch;
    else if (k == "compiles") *value = c->n_compile;
    else if (k == "cache_hits") *value = c->n_cache_hit;
    else if (k == "h2d_bytes") *value = c->h2d;
    else if (k == "d2h_bytes") *value = c->d2h;
    else if (k == "p2p_bytes") *value = c->p2p;
    else if (k == "halo_push_bytes") *value = c->pushed;
    else if (k == "disk_cache_hits") *value = c->n_disk_hit;
    else if (k == "tma_launches") *value = c->n_tma;
    else if (k == "nccl_groups") *value = c->n_nccl_group;           // NCCL send/recv groups issued
    else if (k == "nccl_comm") *value = c->nccl_comm != nullptr;     // an NCCL communicator exists
    else fail(SKL_ERR_INVALID_ARG, "unknown counter " + k);
  });
}

skl_status skl_type_struct(skl_ctx* ctx, const char* name, const char* decl_src, size_t size,
                           size_t align, skl_type* out) {
  return guard([&] {
    Ctx* c = C(ctx);
    if (!name || !decl_src || !out || size == 0) fail(SKL_ERR_INVALID_ARG, "bad struct type");
    for (size_t i = 0; i < c->types.size(); ++i)
      if (c->types[i].name == name) {
        if (c->types[i].decl != decl_src || c->types[i].size != size)
          fail(SKL_ERR_TYPE, std::string("struct type ") + name + " already registered differently");
        *out = (skl_type)i;  // idempotent
        return;
      }
    TypeInfo t;
    t.name = name;
    t.decl = decl_src;
    t.size = size;
    t.align = align ? align : 1;
    c->types.push_back(t);
    *out = (skl_type)(c->types.size() - 1);
  });
}
skl_status skl_type_size(skl_ctx* ctx, skl_type t, size_t* size) {
  return guard([&] {
    if (!size) fail(SKL_ERR_INVALID_ARG, "NULL out");
    *size = C(ctx)->type(t & ~SKL_PTR).size;
  });
}

// ---- containers
skl_status skl_vector_create(skl_ctx* ctx, skl_type t, size_t n, skl_cont** out) {
  return guard([&] {
    if (!out) fail(SKL_ERR_INVALID_ARG, "NULL out");
    *out = wrap(cont_create(C(ctx), t, n, 1, false));
  });
}
skl_status skl_matrix_create(skl_ctx* ctx, skl_type t, size_t rows, size_t cols, skl_cont** out) {
  return guard([&] {
    if (!out) fail(SKL_ERR_INVALID_ARG, "NULL out");
    *out = wrap(cont_create(C(ctx), t, rows, cols, true));
  });
}
skl_status skl_cont_destroy(skl_cont* c) {
  return guard([&] {
    Cont* k = K(c);
    g_cont.erase(k);
    cont_destroy(k);
    c->c = nullptr;
    delete c;
  });
}
skl_status skl_cont_info(skl_cont* c, skl_type* t, size_t* rows, size_t* cols, int* is_matrix) {
  return guard([&] {
    Cont* k = K(c);
    if (t) *t = k->type;
    if (rows) *rows = k->rows;
    if (cols) *cols = k->cols;
    if (is_matrix) *is_matrix = k->matrix;
  });
}
skl_status skl_copy_in(skl_cont* c, const void* host, size_t bytes) {
  return guard([&] {
    Cont* k = K(c);
    if (!host || bytes != k->bytes()) fail(SKL_ERR_SIZE_MISMATCH, "copy_in: byte count must equal the container size");
    materialize_dependents(k);  // deferred readers of the old value run first
    drop_lazy(k);
    if (k->dist.kind == DNONE) {
      void* m = host_mirror(k, SKL_WRITE);
      std::memcpy(m, host, bytes);
    } else {
      host_upload(k, host);
      k->host_valid = false;
    }
  });
}
skl_status skl_copy_out(skl_cont* c, void* host, size_t bytes) {
  return guard([&] {
    Cont* k = K(c);
    if (!host || bytes != k->bytes()) fail(SKL_ERR_SIZE_MISMATCH, "copy_out: byte count must equal the container size");
    if (k->host_valid && k->host) std::memcpy(host, k->host, bytes);
    else host_download(k, host);
  });
}
skl_status skl_copy_out_part(skl_cont* c, int g, void* host, size_t bytes, size_t* first_unit,
                             size_t* nunits) {
  return guard([&] {
    Cont* k = K(c);
    size_t f = 0, n = 0;
    const Range r = core_range(k->units(), k->ctx->G, k->dist, g);
    if (!host || bytes < r.size() * k->unit_bytes()) fail(SKL_ERR_SIZE_MISMATCH, "copy_out_part: buffer too small");
    download_part(k, g, host, &f, &n);
    if (first_unit) *first_unit = f;
    if (nunits) *nunits = n;
  });
}
skl_status skl_host_data(skl_cont* c, int mode, void** host) {
  return guard([&] {
    if (!host || mode < 1 || mode > 3) fail(SKL_ERR_INVALID_ARG, "bad mode or NULL out");
    *host = host_mirror(K(c), mode);
  });
}
skl_status skl_fill(skl_cont* c, const void* value) {
  return guard([&] {
    if (!value) fail(SKL_ERR_INVALID_ARG, "NULL value");
    fill(K(c), value);
  });
}
skl_status skl_set_distribution(skl_cont* c, int kind, int arg, skl_skel* combine) {
  NvtxRange nr("skl_set_distribution");
  return guard([&] {
    Cont* k = K(c);
    Ctx* ctx = k->ctx;
    Dist d{kind, 0};
    switch (kind) {
      case SKL_SINGLE:
        if (arg < 0 || arg >= ctx->G) fail(SKL_ERR_INVALID_ARG, "single: device out of range");
        d.arg = arg;
        break;
      case SKL_COPY:
      case SKL_BLOCK:
        break;
      case SKL_OVERLAP:
        if (arg < 0) fail(SKL_ERR_INVALID_ARG, "overlap size must be >= 0");
        d.arg = arg;
        break;
      default:
        fail(SKL_ERR_INVALID_ARG, "unknown distribution");
    }
    if (combine) {
      if (kind != SKL_COPY) fail(SKL_ERR_DISTRIBUTION, "a combine function needs the copy distribution (A25)");
      Skel* s = S(combine);
      if (s->kind != K_REDUCE || ctx->type(s->tin).size != k->elt)
        fail(SKL_ERR_TYPE, "combine must be a Reduce skeleton over the container's element type");
    }
    materialize(k);  // a deferred Zip/Map result exists before it is moved
    if (!k->dev_valid) {
      k->dist = d;  // data moves lazily (upload at first use)
    } else {
      ensure(k, d, kind == SKL_OVERLAP);
    }
    if (kind == SKL_COPY) k->combine = combine ? S(combine) : nullptr;
  });
}
skl_status skl_get_distribution(skl_cont* c, int* kind, int* arg) {
  return guard([&] {
    Cont* k = K(c);
    if (kind) *kind = k->dist.kind;
    if (arg) *arg = k->dist.arg;
  });
}
skl_status skl_local_part(skl_cont* c, int g, void** dptr, size_t* first_unit, size_t* nunits) {
  return guard([&] {
    Cont* k = K(c);
    if (!dptr) fail(SKL_ERR_INVALID_ARG, "NULL out");
    *dptr = nullptr;
    if (first_unit) *first_unit = 0;
    if (nunits) *nunits = 0;
    if (g < 0 || g >= k->ctx->G || !k->ctx->is_local(g)) return;
    materialize(k);
    // a distribution set on host data becomes resident here (implicit upload)
    if (k->dist.kind != DNONE && !k->dev_valid && k->host_valid) ensure(k, k->dist, k->dist.kind == DOVERLAP);
    sync_ready(k);  // the caller reads the buffer on its own terms: pending chunks first
    Part& p = k->parts[(size_t)g];
    if (!p.ptr || p.valid.empty() || !k->dev_valid) return;
    *dptr = part_ptr(k, g, p.valid.lo);
    if (first_unit) *first_unit = p.valid.lo;
    if (nunits) *nunits = p.valid.size();
  });
}

// ---- skeletons
skl_status skl_map_create(skl_ctx* ctx, const char* src, const char* entry, skl_type in, skl_type out,
                          const skl_type* extra, int nextra, skl_skel** sk) {
  return guard([&] {
    if (!sk || nextra < 0 || (nextra && !extra)) fail(SKL_ERR_INVALID_ARG, "bad arguments");
    *sk = wrap(skel_create(C(ctx), K_MAP, src, entry, in, 0, out, extra, nextra, 0, 0, nullptr));
  });
}
skl_status skl_zip_create(skl_ctx* ctx, const char* src, const char* entry, skl_type left,
                          skl_type right, skl_type out, const skl_type* extra, int nextra,
                          skl_skel** sk) {
  return guard([&] {
    if (!sk || nextra < 0 || (nextra && !extra)) fail(SKL_ERR_INVALID_ARG, "bad arguments");
    *sk = wrap(skel_create(C(ctx), K_ZIP, src, entry, left, right, out, extra, nextra, 0, 0, nullptr));
  });
}
skl_status skl_reduce_create(skl_ctx* ctx, const char* src, const char* entry, skl_type t, skl_skel** sk) {
  return guard([&] {
    if (!sk) fail(SKL_ERR_INVALID_ARG, "NULL out");
    *sk = wrap(skel_create(C(ctx), K_REDUCE, src, entry, t, 0, t, nullptr, 0, 0, 0, nullptr));
  });
}
skl_status skl_scan_create(skl_ctx* ctx, const char* src, const char* entry, skl_type t, skl_skel** sk) {
  return guard([&] {
    if (!sk) fail(SKL_ERR_INVALID_ARG, "NULL out");
    *sk = wrap(skel_create(C(ctx), K_SCAN, src, entry, t, 0, t, nullptr, 0, 0, 0, nullptr));
  });
}
skl_status skl_mapoverlap_create(skl_ctx* ctx, const char* src, const char* entry, skl_type in,
                                 skl_type out, int d, int boundary, const void* neutral, skl_skel** sk) {
  return guard([&] {
    if (!sk) fail(SKL_ERR_INVALID_ARG, "NULL out");
    *sk = wrap(skel_create(C(ctx), K_MAPOVERLAP, src, entry, in, 0, out, nullptr, 0, d, boundary, neutral));
  });
}
skl_status skl_allpairs_create(skl_ctx* ctx, const char* src, const char* entry, skl_type in,
                               skl_type out, skl_skel** sk) {
  return guard([&] {
    if (!sk) fail(SKL_ERR_INVALID_ARG, "NULL out");
    *sk = wrap(allpairs_create(C(ctx), src, entry, nullptr, nullptr, in, out));
  });
}
skl_status skl_allpairs_zr_create(skl_ctx* ctx, const char* zip_src, const char* zip_entry,
                                  const char* reduce_src, const char* reduce_entry, skl_type in,
                                  skl_type out, skl_skel** sk) {
  return guard([&] {
    if (!sk || !reduce_src) fail(SKL_ERR_INVALID_ARG, "NULL out / reduce source");
    *sk = wrap(allpairs_create(C(ctx), zip_src, zip_entry, reduce_src, reduce_entry, in, out));
  });
}
skl_status skl_allpairs_run(skl_skel* sk, skl_cont* a, skl_cont* b, skl_cont** c) {
  NvtxRange nr("skl_allpairs_run");
  return run_out(c, [&](Cont** o) { run_allpairs(S(sk), K(a), K(b), o); });
}
skl_status skl_mapoverlap_bounds(skl_skel* sk, int* proven) {
  return guard([&] {
    Skel* s = S(sk);
    if (s->kind != K_MAPOVERLAP || !proven) fail(SKL_ERR_INVALID_ARG, "not a MapOverlap skeleton / NULL out");
    *proven = s->bounds == 1;
  });
}
skl_status skl_skel_destroy(skl_skel* sk) {
  return guard([&] {
    Skel* s = S(sk);
    g_skel.erase(s);
    skel_destroy(s);
    sk->s = nullptr;
    delete sk;
  });
}
skl_status skl_map_run(skl_skel* sk, skl_cont* in, skl_cont** out, const skl_arg* extra, int nextra) {
  NvtxRange nr("skl_map_run");
  Skel* s = nullptr;
  skl_status st = guard([&] { s = S(sk); K(in); });
  if (st) return st;
  if (s->tout == SKL_VOID) {
    return guard([&] {
      Cont* none = nullptr;
      run_map(s, K(in), &none, extra, nextra);
      if (out) *out = nullptr;
    });
  }
  return run_out(out, [&](Cont** o) { run_map(s, K(in), o, extra, nextra); });
}
skl_status skl_zip_run(skl_skel* sk, skl_cont* left, skl_cont* right, skl_cont** out,
                       const skl_arg* extra, int nextra) {
  NvtxRange nr("skl_zip_run");
  Skel* s = nullptr;
  skl_status st = guard([&] { s = S(sk); K(left); K(right); });
  if (st) return st;
  if (s->tout == SKL_VOID) {
    return guard([&] {
      Cont* none = nullptr;
      run_zip(s, K(left), K(right), &none, extra, nextra);
      if (out) *out = nullptr;
    });
  }
  return run_out(out, [&](Cont** o) { run_zip(s, K(left), K(right), o, extra, nextra); });
}
skl_status skl_reduce_run(skl_skel* sk, skl_cont* in, skl_cont** scalar) {
  NvtxRange nr("skl_reduce_run");
  return run_out(scalar, [&](Cont** o) { run_reduce(S(sk), K(in), o); });
}
skl_status skl_scan_run(skl_skel* sk, skl_cont* in, skl_cont** out) {
  NvtxRange nr("skl_scan_run");
  return run_out(out, [&](Cont** o) { run_scan(S(sk), K(in), o); });
}
skl_status skl_mapoverlap_run(skl_skel* sk, skl_cont* in, skl_cont** out) {
  NvtxRange nr("skl_mapoverlap_run");
  return run_out(out, [&](Cont** o) { run_mapoverlap(S(sk), K(in), o); });
}
skl_status skl_scalar_get(skl_cont* scalar, void* value, size_t bytes) {
  return guard([&] {
    Cont* k = K(scalar);
    if (!value || bytes != k->bytes()) fail(SKL_ERR_SIZE_MISMATCH, "scalar_get: byte count must equal the element size");
    host_download(k, value);
  });
}

// ---- CUDA graphs
struct skl_graph {
  Ctx* ctx;
  int g;
  cudaGraph_t graph;
  cudaGraphExec_t exec;
};
// Several local devices (one process driving every GPU, or logical devices):
// the capture opens on the first device's stream and forks into the other
// devices' streams through an event recorded there, so their calls - and the
// cross-stream barriers between them - are recorded into the same graph; the
// end joins every stream back before closing.  One graph launch then replays
// the multi-device sequence (iterated stencils with their halo exchange): the
// host cost of a call grows with the devices it launches on (~6 us each), more
// than the GPU time of a stencil iteration on 8 GPUs.  Not in the one-process-
// per-GPU mode: its device barriers carry epochs that a replay would repeat.
static std::vector<cudaStream_t> capture_streams(Ctx* c) {
  std::vector<cudaStream_t> out;
  for (int g = c->first_local + 1; g < c->first_local + c->nlocal; ++g) {
    cudaStream_t st = c->D(g).stream;
    bool seen = st == c->D(c->first_local).stream;
    for (cudaStream_t o : out) seen = seen || o == st;
    if (!seen) out.push_back(st);
  }
  return out;
}
static int stream_device(Ctx* c, cudaStream_t st) {
  for (int g = c->first_local; g < c->first_local + c->nlocal; ++g)
    if (c->D(g).stream == st) return c->D(g).phys;
  return c->D(c->first_local).phys;
}
skl_status skl_capture_begin(skl_ctx* ctx) {
  return guard([&] {
    Ctx* c = C(ctx);
    if (c->dist_mode) fail(SKL_ERR_UNSUPPORTED, "graph capture in the one-process-per-GPU mode");
    if (c->capturing) fail(SKL_ERR_INVALID_ARG, "already capturing");
    c->set_device(c->first_local);
    cudaStream_t origin = c->D(c->first_local).stream;
    SKL_CUDA(cudaStreamBeginCapture(origin, cudaStreamCaptureModeRelaxed));
    c->capturing = true;
    const auto others = capture_streams(c);
    if (!others.empty()) {
      if (!c->cap_fork) SKL_CUDA(cudaEventCreateWithFlags(&c->cap_fork, cudaEventDisableTiming));
      SKL_CUDA(cudaEventRecord(c->cap_fork, origin));
      for (cudaStream_t st : others) {
        SKL_CUDA(cudaSetDevice(stream_device(c, st)));
        SKL_CUDA(cudaStreamWaitEvent(st, c->cap_fork, 0));
      }
      c->set_device(c->first_local);
    }
  });
}
skl_status skl_capture_end(skl_ctx* ctx, skl_graph** out) {
  return guard([&] {
    Ctx* c = C(ctx);
    if (!c->capturing || !out) fail(SKL_ERR_INVALID_ARG, "not capturing / NULL out");
    c->capturing = false;
    cudaStream_t origin = c->D(c->first_local).stream;
    const auto others = capture_streams(c);
    if (c->cap_join.size() < others.size()) c->cap_join.resize(others.size(), nullptr);
    for (size_t i = 0; i < others.size(); ++i) {
      const int dev = stream_device(c, others[i]);
      SKL_CUDA(cudaSetDevice(dev));
      if (!c->cap_join[i]) SKL_CUDA(cudaEventCreateWithFlags(&c->cap_join[i], cudaEventDisableTiming));
      SKL_CUDA(cudaEventRecord(c->cap_join[i], others[i]));
      c->set_device(c->first_local);
      SKL_CUDA(cudaStreamWaitEvent(origin, c->cap_join[i], 0));
    }
    c->set_device(c->first_local);
    cudaGraph_t graph = nullptr;
    SKL_CUDA(cudaStreamEndCapture(origin, &graph));
    cudaGraphExec_t exec = nullptr;
    cudaError_t e = cudaGraphInstantiate(&exec, graph, 0);
    if (e != cudaSuccess) {
      cudaGraphDestroy(graph);
      cuda_check(e, "cudaGraphInstantiate");
    }
    *out = new skl_graph{c, c->first_local, graph, exec};
  });
}
skl_status skl_graph_launch(skl_graph* gr) {
  return guard([&] {
    if (!gr) fail(SKL_ERR_INVALID_ARG, "NULL graph");
    Ctx* c = gr->ctx;
    if (c->capturing) fail(SKL_ERR_INVALID_ARG, "graph launch while capturing");
    cudaStream_t origin = c->D(gr->g).stream;
    // a multi-device graph runs after the work already queued on every device
    // stream, and later work on any of them runs after it
    const auto others = capture_streams(c);
    if (c->cap_join.size() < others.size()) c->cap_join.resize(others.size(), nullptr);
    for (size_t i = 0; i < others.size(); ++i) {
      SKL_CUDA(cudaSetDevice(stream_device(c, others[i])));
      if (!c->cap_join[i]) SKL_CUDA(cudaEventCreateWithFlags(&c->cap_join[i], cudaEventDisableTiming));
      SKL_CUDA(cudaEventRecord(c->cap_join[i], others[i]));
      c->set_device(gr->g);
      SKL_CUDA(cudaStreamWaitEvent(origin, c->cap_join[i], 0));
    }
    c->set_device(gr->g);
    SKL_CUDA(cudaGraphLaunch(gr->exec, origin));
    c->n_launch += 1;
    if (!others.empty()) {
      if (!c->cap_fork) SKL_CUDA(cudaEventCreateWithFlags(&c->cap_fork, cudaEventDisableTiming));
      SKL_CUDA(cudaEventRecord(c->cap_fork, origin));
      for (cudaStream_t st : others) {
        SKL_CUDA(cudaSetDevice(stream_device(c, st)));
        SKL_CUDA(cudaStreamWaitEvent(st, c->cap_fork, 0));
      }
      c->set_device(gr->g);
    }
  });
}
skl_status skl_graph_destroy(skl_graph* gr) {
  return guard([&] {
    if (!gr) return;
    cudaGraphExecDestroy(gr->exec);
    cudaGraphDestroy(gr->graph);
    delete gr;
  });
}

// ---- offline compilation / introspection
skl_status skl_init_offline(skl_ctx** out) {
  return guard([&] {
    if (!out) fail(SKL_ERR_INVALID_ARG, "NULL out");
    Ctx* c = ctx_create_offline();
    *out = new skl_ctx{c};
    g_ctx[c] = *out;
  });
}
skl_status skl_skel_cubin(skl_skel* sk, void* buf, size_t cap, size_t* size) {
  return guard([&] {
    Skel* s = S(sk);
    if (!size) fail(SKL_ERR_INVALID_ARG, "NULL size");
    *size = s->prog->cubin.size();
    if (buf && cap >= *size) std::memcpy(buf, s->prog->cubin.data(), *size);
  });
}
skl_status skl_skel_source(skl_skel* sk, char* buf, size_t cap, size_t* size) {
  return guard([&] {
    Skel* s = S(sk);
    if (!size) fail(SKL_ERR_INVALID_ARG, "NULL size");
    *size = s->prog->source.size() + 1;
    if (buf && cap >= *size) std::memcpy(buf, s->prog->source.c_str(), *size);
  });
}

// ---- host-only planning
skl_status skl_plan_range(size_t units, int G, int kind, int arg, int g, int with_halo, size_t* lo,
                          size_t* hi) {
  return guard([&] {
    if (G < 1 || g < 0 || g >= G || !lo || !hi) fail(SKL_ERR_INVALID_ARG, "bad arguments");
    const Dist d{kind, arg};
    const Range r = with_halo ? need_range(units, G, d, g) : core_range(units, G, d, g);
    *lo = r.lo;
    *hi = r.hi;
  });
}
skl_status skl_plan_transfers(size_t units, int G, int from_kind, int from_arg, int to_kind, int to_arg,
                              int64_t* tuples, size_t cap, size_t* ntransfers) {
  return guard([&] {
    if (G < 1 || !ntransfers) fail(SKL_ERR_INVALID_ARG, "bad arguments");
    const std::vector<Transfer> tr = plan_transfers(units, G, Dist{from_kind, from_arg}, from_kind == SKL_OVERLAP,
                                                    Dist{to_kind, to_arg}, to_kind == SKL_OVERLAP);
    *ntransfers = tr.size();
    for (size_t i = 0; i < tr.size() && i < cap && tuples; ++i) {
      tuples[5 * i + 0] = tr[i].src;
      tuples[5 * i + 1] = (int64_t)tr[i].src_unit;
      tuples[5 * i + 2] = tr[i].dst;
      tuples[5 * i + 3] = (int64_t)tr[i].dst_unit;
      tuples[5 * i + 4] = (int64_t)tr[i].n;
    }
  });
}

}  // extern "C"
