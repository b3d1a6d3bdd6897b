// skeletons.cpp — skeleton objects and their executors (SURVEY §1 layer B5).
//
// A skeleton is "a higher-order function that executes one or more
// user-defined (so-called customizing) functions in a pre-defined parallel
// manner".  Creation compiles the customising source into the
// skeleton's sm_100a kernel template (NVRTC, compiler.cpp); a call
// ("resultVector = neg(inputVector)") makes the inputs resident in
// the distribution the skeleton needs (implicit transfers / redistribution,
// container.cpp), launches one kernel per device on that device's part, and
// performs the one cross-device step the skeleton has, if any:
//   Map, Zip      none                       (block: independent parts)
//   Reduce        ordered fold of the G device partials
//   Scan          device totals -> carry-in of the later devices
//   MapOverlap    overlap halo refresh before the stencil
#include <functional>
#include <algorithm>
#include <cstdio>
#include <numeric>

#include <cuda.h>
#include <cudaTypedefs.h>

#include "skl_internal.h"

namespace skl {
struct alignas(64) SklTensorMap {
  unsigned char b[128];
};
static_assert(sizeof(SklTensorMap) == sizeof(CUtensorMap), "tensor map size");
}  // namespace skl

namespace skl {

extern void set_last_error(const std::string& s);

namespace {

size_t gcd_sz(size_t a, size_t b) { return b ? gcd_sz(b, a % b) : a; }
size_t lcm_sz(size_t a, size_t b) { return a / gcd_sz(a, b) * b; }
// elements per chunk so that VEC * size is a multiple of 16 bytes for every size
size_t vec_for(std::initializer_list<size_t> sizes) {
  size_t v = 1;
  for (size_t s : sizes)
    if (s) v = lcm_sz(v, 16 / gcd_sz(16, s));
  return v;
}
bool aligned16(const void* p) { return ((uintptr_t)p & 15u) == 0; }
size_t ceil_div(size_t a, size_t b) { return (a + b - 1) / b; }

std::string defs_common(Ctx* ctx, const std::string& entry, int block) {
  std::string s;
  s += "#define SKL_BLOCK " + std::to_string(block) + "\n";
  s += "#define SKL_CBLOCK " + std::to_string(kCombineBlock) + "\n";
  s += "#define SKL_DEBUG_BOUNDS " + std::to_string(ctx->debug_bounds ? 1 : 0) + "\n";
  s += "#define SKL_FUNC " + entry + "\n";
  return s;
}

std::string tname(Ctx* ctx, int t) { return ctx->type(t).name; }
// rows per thread, tile rows, tiles per block; a block of 2+ tiles marks a heavy
// function (>= 64 registers), which also gets the unguarded full-tile path
// (option mo_full: 1 / 0 forces it on / off)
std::string mo_rows_defs(Ctx* ctx, int rh, int th, int kt, int force_full = -1) {
  const bool full = force_full >= 0 ? force_full == 1 : ctx->mo_full >= 0 ? ctx->mo_full == 1 : kt > 1;
  return "#define SKL_RH " + std::to_string(rh) + "\n#define SKL_TH " + std::to_string(th) + "\n#define SKL_MO_KT " +
         std::to_string(kt) + "\n#define SKL_MO_HEAVY " + (full ? "1" : "0") + "\n";
}

// Scratch buffer per (skeleton, device), grown on demand.
void* scratch(Skel* s, std::map<int, Scratch>& m, int g, size_t bytes, bool zero) {
  Scratch& sc = m[g];
  if (sc.bytes < bytes) {
    if (sc.ptr) device_free(s->ctx, g, sc.ptr);
    sc.ptr = device_alloc(s->ctx, g, bytes);
    sc.bytes = bytes;
    if (zero) {
      s->ctx->set_device(g);
      SKL_CUDA(cudaMemsetAsync(sc.ptr, 0, bytes, s->ctx->D(g).stream));
    }
  }
  return sc.ptr;
}

}  // namespace

// ------------------------------------------------------------------ creation
Skel* skel_create(Ctx* ctx, int kind, const char* src, const char* entry, int tin, int tin2,
                  int tout, const int* extra, int nextra, int d, int boundary, const void* neutral) {
  if (!src) fail(SKL_ERR_INVALID_ARG, "customising function source is NULL");
  auto s = std::make_unique<Skel>();
  std::function<std::string(int, int)> mo_geo;  // MapOverlap: register-block defines
  std::string mo_tail;                          // MapOverlap: defines after the geometry
  s->ctx = ctx;
  s->kind = kind;
  s->user_src = src;
  s->entry = (entry && *entry) ? std::string(entry) : detect_entry(s->user_src);
  s->tin = tin;
  s->tin2 = tin2;
  s->tout = tout;
  for (int i = 0; i < nextra; ++i) s->extra.push_back(extra[i]);
  s->d = d;
  s->boundary = boundary;
  const std::string user = "\n// ---- customising function (user source)\n#line 1 \"user_source\"\n" +
                           s->user_src + "\n#line 1 \"skeleton_template\"\n";
  // launch geometry is fixed at creation (compiled into the program)
  s->block = ctx->block_threads;
  s->unroll = ctx->map_unroll;
  // Map / Zip over a function with a loop: interleaved, one element per lane
  const bool auto_il = (kind == K_MAP || kind == K_ZIP) && ctx->map_interleave == 0 && ctx->map_auto &&
                       has_loop(s->user_src);
  s->interleave = ctx->map_interleave != 0 || auto_il;
  std::string defs = defs_common(ctx, s->entry, s->block);
  std::string body;
  switch (kind) {
    case K_MAP:
    case K_ZIP: {
      const size_t si = ctx->type(tin).size;
      const size_t si2 = kind == K_ZIP ? ctx->type(tin2).size : 0;
      const size_t so = tout == SKL_VOID ? 0 : ctx->type(tout).size;
      if (si == 0 || (kind == K_ZIP && si2 == 0)) fail(SKL_ERR_TYPE, "void input type");
      const size_t vec = std::min<size_t>(vec_for({si, si2, so}), 64);
      defs += "#define SKL_TIN " + tname(ctx, tin) + "\n";
      if (kind == K_ZIP) defs += "#define SKL_TIN2 " + tname(ctx, tin2) + "\n#define SKL_ZIP 1\n";
      else defs += "#define SKL_ZIP 0\n";
      if (tout == SKL_VOID) defs += "#define SKL_TOUT void\n#define SKL_OUT_VOID 1\n";
      else defs += "#define SKL_TOUT " + tname(ctx, tout) + "\n#define SKL_OUT_VOID 0\n";
      defs += "#define SKL_VEC " + std::to_string(vec) + "\n";
      defs += "#define SKL_UNROLL " + std::to_string(ctx->map_unroll) + "\n";
      s->ilj = ctx->map_il_elems > 0 ? ctx->map_il_elems : (auto_il ? 1 : (int)(ctx->map_unroll * vec));
      defs += "#define SKL_ILJ " + std::to_string(s->ilj) + "\n";
      std::string xp, xa;
      for (size_t k = 0; k < s->extra.size(); ++k) {
        const int t = s->extra[k];
        const bool ptr = (t & SKL_PTR) != 0;
        const int base = t & ~SKL_PTR;
        if (ctx->type(base).size == 0) fail(SKL_ERR_TYPE, "void extra argument");
        xp += ", " + tname(ctx, base) + (ptr ? "* " : " ") + "skl_x" + std::to_string(k);
        xa += ", skl_x" + std::to_string(k);
      }
      defs += "#define SKL_XPARAMS " + xp + "\n#define SKL_XARGS " + xa + "\n";
      body = user + kernel_template("common.cuh") + kernel_template("map.cuh");
      break;
    }
    case K_REDUCE:
    case K_SCAN: {
      const size_t st = ctx->type(tin).size;
      if (st == 0) fail(SKL_ERR_TYPE, "void element type");
      defs += "#define SKL_T " + tname(ctx, tin) + "\n";
      const int rvec = (16 % st == 0) ? (int)(16 / st) : 1;
      defs += "#define SKL_RVEC " + std::to_string(rvec) + "\n#define SKL_RU 4\n";
      if (kind == K_SCAN) {
        // 8 chunks (128 B) per thread: 8192 fp32 elements per tile (SURVEY §7 hard part 2)
        const int ch = (16 % st == 0) ? ctx->scan_chunks : 0;
        s->scan_ch = ch;
        const int items = ch ? (int)(ch * 16 / st) : 8;
        defs += "#define SKL_CH " + std::to_string(ch) + "\n#define SKL_ITEMS " + std::to_string(items) + "\n";
        defs += std::string("#define SKL_PACKED ") + (st <= 4 ? "1" : "0") + "\n";
        defs += "#define SKL_SCAN_VARIANT " + std::to_string(ctx->scan_variant) + "\n";
        s->scan_sub = ctx->scan_sub;
        s->scan_variant = ctx->scan_variant;
        s->scan_fstride = ctx->scan_fstride;
        defs += "#define SKL_FSTRIDE " + std::to_string(s->scan_fstride) + "\n";
        defs += "#define SKL_SPIN_NS " + std::to_string(ctx->scan_spin_ns) + "\n";
        defs += "#define SKL_MINB " + std::to_string(ctx->scan_minb) + "\n";
        defs += "#define SKL_MINB_P " + std::to_string(ctx->scan_minb_pipe) + "\n";
        defs += "#define SKL_LBW " + std::to_string(ctx->scan_lbw) + "\n";
        defs += "#define SKL_SUB " + std::to_string(s->scan_sub) + "\n";
      }
      s->cunr = ctx->combine_unroll > 0 ? ctx->combine_unroll : 2;
      defs += "#define SKL_CUNR " + std::to_string(s->cunr) + "\n";
      body = user + kernel_template("common.cuh") + kernel_template("op.cuh") +
             kernel_template("reduce.cuh") + (kind == K_SCAN ? kernel_template("scan.cuh") : "");
      break;
    }
    case K_MAPOVERLAP: {
      const size_t si = ctx->type(tin).size, so = ctx->type(tout).size;
      if (si == 0 || so == 0) fail(SKL_ERR_TYPE, "MapOverlap needs non-void types");
      if (16 % si != 0) fail(SKL_ERR_TYPE, "MapOverlap element size must divide 16 bytes");
      if (d < 0) fail(SKL_ERR_INVALID_ARG, "negative overlap size");
      if (boundary != SKL_NEUTRAL && boundary != SKL_NEAREST) fail(SKL_ERR_INVALID_ARG, "bad boundary mode");
      {
        // static get() bounds (P:L366-368 future work): reject provable violations
        // now; proven functions need no runtime check even in debug mode
        std::string why;
        s->bounds = check_get_bounds(s->user_src, d, &why);
        if (s->bounds < 0) fail(SKL_ERR_OUT_OF_RANGE, "static get() check (P:L362-368): " + why);
        if (s->bounds == 1 && ctx->debug_bounds) {
          const std::string on = "#define SKL_DEBUG_BOUNDS 1\n", off = "#define SKL_DEBUG_BOUNDS 0\n";
          const size_t at = defs.find(on);
          if (at != std::string::npos) defs.replace(at, on.size(), off);
        }
      }
      s->neutral.assign(si, 0);
      if (neutral) std::memcpy(s->neutral.data(), neutral, si);
      const int epc = (int)(16 / si);
      const int A = (int)ceil_div((size_t)d, (size_t)epc) * epc;
      // default register block: one 16-byte-wide run of outputs per row; 8 rows
      // for wider elements, and for byte images 4 rows unless the function then
      // spills at the 64-register budget (checked after compiling, below: then
      // 2 rows).  Swept on B200 (tools/mo_probe.py, profiles/sweeps): identity u8
      // 30.8 -> 26.6 us at 4 rows, the separable Sobel 75.9 -> 72.7 us, while
      // Listing 1.5's Sobel (IEEE sqrtf subroutine) spills at 4 rows (77 -> 92 us);
      // Gaussian f32 at 8 rows / <= 128 registers.
      int cw = (int)(16 / std::min<size_t>(so, 16) > 0 ? 16 / std::min<size_t>(so, 16) : 1);
      int rh = si >= 4 ? 8 : (si == 1 ? 4 : 2);
      if (ctx->mo_cw > 0) cw = ctx->mo_cw;  // register block per thread (tuning knobs)
      if (ctx->mo_rh > 0) rh = ctx->mo_rh;
      s->mo_auto_rh = ctx->mo_rh == 0 && si == 1;
      // byte images, geometry fully automatic: a heavy function gets the 8 x 8
      // register block below (chosen after compiling)
      s->mo_auto_byte = si == 1 && ctx->mo_rh == 0 && ctx->mo_cw == 0 && ctx->mo_kt == 0 && ctx->mo_full < 0;
      const int nthr = ctx->block_threads;
      const std::string pre = defs;
      // the register-block geometry's defines (and the skeleton's copy of it)
      mo_geo = [&, pre, nthr, A, si, so, tin, tout, d, boundary](int cw_, int rh_) {
        if ((cw_ * (int)si) % 16 != 0 && (16 % (cw_ * (int)si)) != 0)
          fail(SKL_ERR_INVALID_ARG, "mo_cw x element size must divide or be a multiple of 16 bytes");
        const int tw = 32 * cw_;
        const int rows_thr = nthr / 32;
        int th = rows_thr * rh_;
        while (rh_ > 1 && (size_t)(th + 2 * d) * (size_t)(tw + 2 * A) * si > 44 * 1024) {
          rh_ /= 2;
          th = rows_thr * rh_;
        }
        s->mo_tw = tw;
        s->mo_a = A;
        s->mo_pitch = tw + 2 * A;
        s->mo_cw = cw_;
        s->mo_rh = rh_;
        s->mo_th = th;
        std::string g = pre;
        g += "#define SKL_TIN " + tname(ctx, tin) + "\n#define SKL_TOUT " + tname(ctx, tout) + "\n";
        g += "#define SKL_D " + std::to_string(d) + "\n#define SKL_BOUNDARY " + std::to_string(boundary) + "\n";
        g += "#define SKL_A " + std::to_string(A) + "\n";
        g += "#define SKL_PITCH " + std::to_string(tw + 2 * A) + "\n";
        g += "#define SKL_TW " + std::to_string(tw) + "\n#define SKL_CW " + std::to_string(cw_) + "\n";
        g += "#define SKL_OUTB " + std::to_string((size_t)cw_ * so) + "\n#define SKL_SO " + std::to_string(so) + "\n";
        g += "#define SKL_MO1D 0\n";
        return g;
      };
      defs = mo_geo(cw, rh);
      // resident blocks per SM the register allocation must allow (default: 64
      // registers per thread for byte images - 87 registers halved the Sobel
      // occupancy and cost 30 % - and 128 for wider elements)
      const int minb = ctx->mo_minb > 0 ? ctx->mo_minb : std::max(1, 65536 / (nthr * (si >= 4 ? 128 : 64)));
      defs += "#define SKL_MO_MINB " + std::to_string(minb) + "\n";
      // the TMA / warp-specialised kernel (one extra producer warp) keeps the same
      // per-thread register budget
      const int wsminb =
          ctx->mo_ws_minb > 0 ? ctx->mo_ws_minb : std::max(1, 65536 / ((nthr + 32) * (si >= 4 ? 128 : 64)));
      defs += "#define SKL_WS_MINB " + std::to_string(wsminb) + "\n";
      mo_tail = "#define SKL_MO_MINB " + std::to_string(minb) + "\n#define SKL_WS_MINB " + std::to_string(wsminb) + "\n";
      s->mo_kt = ctx->mo_kt > 0 ? ctx->mo_kt : 1;
      s->mo_defs = defs;  // rows and tiles per block go in last (mo_rows_defs): chosen after compiling
      defs += mo_rows_defs(ctx, s->mo_rh, s->mo_th, s->mo_kt);
      body = user + kernel_template("common.cuh") + kernel_template("mapoverlap.cuh");
      // 1-D variant (vector containers), compiled lazily in run_mapoverlap
      break;
    }
    default:
      fail(SKL_ERR_INVALID_ARG, "unknown skeleton kind");
  }
  std::string log;
  s->prog = compile(ctx, defs + program_source(ctx, body), &log);
  if (kind == K_MAPOVERLAP && !ctx->offline) {
    // geometry chosen after compiling, from the TMA tile kernel's resources
    // (tools/mo_probe.py on B200):
    //  * tiles per block (mo_kt = 0): 2 for functions that need >= 64 registers -
    //    the second tile's copy lands while f runs on the first - else 1
    //    (Gaussian 127 -> 117 us, separable Sobel 69.6 -> 65.6 us at 2 tiles;
    //    identity u8 26.7 us at 1 vs 28.7 at 2);
    //  * byte images: 4 rows per thread unless the kernel then needs more local
    //    memory than the 16-byte call frame of the IEEE sqrt subroutine (spills
    //    at the 64-register budget: Listing 1.5's Sobel at 4 rows and 1 tile,
    //    77 -> 92 us), else 2 rows.
    auto attrs = [&](cudaFuncAttributes* fa) {
      ctx->set_device(ctx->first_local);
      cudaKernel_t k = nullptr;
      if (cudaLibraryGetKernel(&k, s->prog->lib, "skl_mo2d_t") == cudaSuccess &&
          cudaFuncGetAttributes(fa, (const void*)k) == cudaSuccess)
        return true;
      (void)cudaGetLastError();
      return false;
    };
    auto recompile = [&](int rh, int kt) {
      s->mo_th = s->mo_th / s->mo_rh * rh;
      s->mo_rh = rh;
      s->mo_kt = kt;
      s->prog = compile(ctx, s->mo_defs + mo_rows_defs(ctx, rh, s->mo_th, kt) + program_source(ctx, body), &log);
    };
    cudaFuncAttributes fa{};
    if (attrs(&fa) && s->mo_auto_byte && fa.numRegs >= 64) {
      //  * byte images with a heavy function (every option automatic): 8 x 8
      //    outputs per thread, one tile per block, the unguarded full-tile loop
      //    (bench context, 8192^2: Listing 1.5 67.6 -> 65.6 us, the tuned Sobel
      //    51.2 -> 47.1 us; profiles/sweeps/sweep_r02_sobel.log r10)
      s->mo_defs = mo_geo(8, 8) + mo_tail;
      s->mo_kt = 1;
      s->prog = compile(ctx, s->mo_defs + mo_rows_defs(ctx, s->mo_rh, s->mo_th, 1, 1) + program_source(ctx, body),
                        &log);
    } else if (attrs(&fa)) {
      const bool heavy = fa.numRegs >= 64;
      if (ctx->mo_kt == 0 && heavy) {
        recompile(s->mo_rh, 2);
        if (!attrs(&fa)) fa.localSizeBytes = 0;
      }
      if (s->mo_auto_rh && s->mo_rh > 2 && fa.localSizeBytes > 16) recompile(2, s->mo_kt);
    }
  }
  Skel* raw = s.release();
  ctx->skels.insert(raw);
  return raw;
}

void skel_destroy(Skel* s) {
  Ctx* ctx = s->ctx;
  // deferred results of this skeleton must exist before it goes away
  for (Cont* c : std::vector<Cont*>(ctx->conts.begin(), ctx->conts.end()))
    if (c->lazy.s == s) materialize(c);
  for (Skel* k : ctx->skels) {
    k->fused.erase(s);
    k->composed.erase(s);
  }
  for (auto* m : {&s->scratch_red, &s->scratch_scan, &s->scratch_stage})
    for (auto& kv : *m)
      if (kv.second.ptr && ctx->is_local(kv.first)) device_free(ctx, kv.first, kv.second.ptr);
  for (Cont* c : ctx->conts)
    if (c->combine == s) c->combine = nullptr;
  ctx->skels.erase(s);
  delete s;
}

// ------------------------------------------------------------------ helpers
namespace {

Dist default_dist(Cont* c, Dist def) { return c->dist.kind == DNONE ? def : c->dist; }
// elementwise skeletons compute a container's core: overlap behaves as block
Dist elementwise(Dist d) { return d.kind == DOVERLAP ? Dist{DBLOCK, 0} : d; }

Cont* output_for(Ctx* ctx, Cont** out, int type, size_t rows, size_t cols, bool matrix) {
  if (*out) {
    Cont* o = *out;
    if (o->type != type) fail(SKL_ERR_TYPE, "output container has the wrong element type");
    if (o->rows != rows || o->cols != cols) fail(SKL_ERR_SIZE_MISMATCH, "output container has the wrong size");
    return o;
  }
  *out = cont_create(ctx, type, rows, cols, matrix);
  return *out;
}

struct ExtraArgs {
  std::vector<std::vector<unsigned char>> scalars;
  std::vector<Cont*> conts;
  std::vector<int> modes;
};

ExtraArgs prepare_extras(Skel* s, const skl_arg* extra, int nextra) {
  if (nextra != (int)s->extra.size())
    fail(SKL_ERR_INVALID_ARG, "skeleton expects " + std::to_string(s->extra.size()) + " extra arguments");
  ExtraArgs ea;
  ea.scalars.resize((size_t)nextra);
  ea.conts.assign((size_t)nextra, nullptr);
  ea.modes.assign((size_t)nextra, 0);
  for (int k = 0; k < nextra; ++k) {
    const int t = s->extra[(size_t)k];
    const bool ptr = (t & SKL_PTR) != 0;
    const size_t sz = s->ctx->type(t & ~SKL_PTR).size;
    if (ptr) {
      if (extra[k].kind != SKL_ARG_CONT || !extra[k].cont || !extra[k].cont->c)
        fail(SKL_ERR_INVALID_ARG, "extra argument " + std::to_string(k) + " must be a container");
      Cont* c = extra[k].cont->c;
      if (c->elt != sz) fail(SKL_ERR_TYPE, "extra container argument has the wrong element type");
      // A27: a container argument is read at arbitrary indices: every device needs
      // the whole container, i.e. the copy distribution.
      ensure(c, Dist{DCOPY, 0}, false);
      if (extra[k].mode & SKL_WRITE) materialize_dependents(c);  // c changes in place
      ea.conts[(size_t)k] = c;
      ea.modes[(size_t)k] = extra[k].mode ? extra[k].mode : SKL_READ;
    } else {
      if (extra[k].kind != SKL_ARG_SCALAR || !extra[k].value || extra[k].bytes != sz)
        fail(SKL_ERR_INVALID_ARG, "extra argument " + std::to_string(k) + " must be a scalar of " +
                                      std::to_string(sz) + " bytes");
      ea.scalars[(size_t)k].assign((const unsigned char*)extra[k].value,
                                   (const unsigned char*)extra[k].value + sz);
    }
  }
  return ea;
}

void finish_extras(Ctx* ctx, ExtraArgs& ea, int ndev_exec) {
  for (size_t k = 0; k < ea.conts.size(); ++k) {
    Cont* c = ea.conts[k];
    if (!c || !(ea.modes[k] & SKL_WRITE)) continue;
    c->host_valid = false;
    // replicas written independently (A25); one device: its replica is the fold
    if (ctx->G > 1 && ndev_exec >= 1) c->diverged = true;
  }
}

}  // namespace

// ------------------------------------------------------------------ Map / Zip
// Lazy fusion of chains: a Map g applied to the deferred
// result of a Map/Zip f becomes one elementwise skeleton computing g(f(x[, y]))
// (both sources renamed by macros: both may be called `func`).  Compiled once
// per (g, f) pair; nullptr if it cannot be composed (types differ, or the two
// sources clash), and the call then runs eagerly.
static Skel* composed_skel(Skel* g, Skel* f) {
  auto it = g->composed.find(f);
  if (it != g->composed.end()) return it->second;
  Ctx* ctx = g->ctx;
  Skel* c = nullptr;
  if (g->kind == K_MAP && g->extra.empty() && f->extra.empty() && g->tin == f->tout &&
      (f->kind == K_MAP || f->kind == K_ZIP) && f->tout != SKL_VOID && g->tout != SKL_VOID) {
    const std::string id = "skl_c" + std::to_string(++ctx->composed_id);
    const bool zip = f->kind == K_ZIP;
    std::string src = "#define " + f->entry + " " + id + "_f\n" + f->user_src + "\n#undef " + f->entry + "\n";
    src += "#define " + g->entry + " " + id + "_g\n" + g->user_src + "\n#undef " + g->entry + "\n";
    src += tname(ctx, g->tout) + " " + id + "(" + tname(ctx, f->tin) + " x" +
           (zip ? ", " + tname(ctx, f->tin2) + " y" : std::string()) + ") { return " + id + "_g(" + id +
           "_f(x" + (zip ? ", y" : "") + ")); }\n";
    try {
      c = skel_create(ctx, f->kind, src.c_str(), id.c_str(), f->tin, f->tin2, g->tout, nullptr, 0, 0, 0,
                      nullptr);
    } catch (const Error&) {
      c = nullptr;  // e.g. a helper function defined in both sources
    }
  }
  g->composed[f] = c;
  return c;
}

static void run_elementwise(Skel* s, Cont* in, Cont* in2, Cont** out, const skl_arg* extra,
                            int nextra) {
  Ctx* ctx = s->ctx;
  if (in->type != s->tin && in->elt != ctx->type(s->tin).size)
    fail(SKL_ERR_TYPE, "input container type does not match the skeleton");
  if (in2) {
    if (in2->elt != ctx->type(s->tin2).size) fail(SKL_ERR_TYPE, "right input type mismatch");
    if (in2->rows * in2->cols != in->rows * in->cols || in2->rows != in->rows)
      fail(SKL_ERR_SIZE_MISMATCH, "zip inputs differ in size (P:L257-259)");
  }
  if (!in2 && nextra == 0 && in->lazy.s && ctx->lazy_fusion && s->kind == K_MAP) {
    if (Skel* c = composed_skel(s, in->lazy.s)) {
      const Lazy L = in->lazy;
      if (*out == nullptr) {
        // stays deferred: g(f(...)) of f's inputs
        Cont* o = cont_create(ctx, s->tout, in->rows, in->cols, in->matrix);
        o->lazy = Lazy{c, L.l, L.r, L.d};
        o->dist = L.d;
        L.l->dependents.push_back(o);
        if (L.r && L.r != L.l) L.r->dependents.push_back(o);
        *out = o;
        return;
      }
      // an explicit output: one kernel from f's inputs, no intermediate
      run_elementwise(c, L.l, L.r, out, nullptr, 0);
      return;
    }
  }
  const Dist din = elementwise(default_dist(in, Dist{DBLOCK, 0}));  // A6
  // keep_ready: chunks of an upload still in flight are consumed one by one below
  ensure(in, in->dist.kind == DOVERLAP ? in->dist : din, false, /*keep_ready=*/true);
  if (in2) {
    // A7: the right input follows the left input's distribution
    if (!(elementwise(in2->dist) == din && in2->dev_valid)) ensure(in2, din, false);
    else ensure(in2, in2->dist, false);
  }
  if (*out == nullptr && nextra == 0 && s->tout != SKL_VOID && ctx->lazy_fusion &&
      in->dist.kind != DOVERLAP && (!in2 || in2->dist.kind != DOVERLAP)) {
    // deferred (lazy fusion): nothing runs until the result is used
    Cont* o = cont_create(ctx, s->tout, in->rows, in->cols, in->matrix);
    o->lazy = Lazy{s, in, in2, din};
    o->dist = din;
    in->dependents.push_back(o);
    if (in2 && in2 != in) in2->dependents.push_back(o);
    *out = o;
    return;
  }
  ExtraArgs ea = prepare_extras(s, extra, nextra);
  // the input's pending upload chunks (chunked copy_in / upload on first use):
  // one launch per chunk, each waiting only for its own chunk
  std::vector<std::vector<Ready>> chunks((size_t)ctx->G);
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) {
    chunks[(size_t)g].swap(in->parts[(size_t)g].ready);
    std::sort(chunks[(size_t)g].begin(), chunks[(size_t)g].end(),
              [](const Ready& a, const Ready& b) { return a.r.lo < b.r.lo; });
  }
  Cont* o = nullptr;
  if (s->tout != SKL_VOID) {
    o = output_for(ctx, out, s->tout, in->rows, in->cols, in->matrix);
    if (o == in && !(in->dist == din)) fail(SKL_ERR_INVALID_ARG, "in-place call needs a block/copy/single input");
    prepare_output(o, din, 0);
  }
  const size_t vec = std::min<size_t>(
      vec_for({ctx->type(s->tin).size, in2 ? ctx->type(s->tin2).size : 0,
               s->tout == SKL_VOID ? 0 : ctx->type(s->tout).size}), 64);
  const size_t per_block = (size_t)s->block * (size_t)s->unroll;
  int ndev = 0;
  auto launch_range = [&](int g, const Range& r) {
    const void* pin = part_ptr(in, g, r.lo);
    const void* pin2 = in2 ? part_ptr(in2, g, r.lo) : nullptr;
    void* pout = o ? part_ptr(o, g, r.lo) : nullptr;
    unsigned long long n = (unsigned long long)(r.size() * in->cols);
    const bool vec_ok = aligned16(pin) && (!in2 || aligned16(pin2)) && (!o || aligned16(pout));
    std::vector<void*> args;
    args.push_back(&pin);
    if (in2) args.push_back(&pin2);
    args.push_back(&pout);
    args.push_back(&n);
    std::vector<void*> xptr(ea.conts.size(), nullptr);
    for (size_t k = 0; k < ea.conts.size(); ++k) {
      if (ea.conts[k]) {
        xptr[k] = part_ptr(ea.conts[k], g, 0);
        args.push_back(&xptr[k]);
      } else {
        args.push_back(ea.scalars[k].data());
      }
    }
    size_t grid;
    const char* kname;
    if (s->interleave) {
      grid = std::max<size_t>(1, ceil_div(n, (size_t)s->block * (size_t)s->ilj));
      kname = "skl_map_il";
    } else if (vec_ok) {
      grid = std::max<size_t>(1, ceil_div(n / vec, per_block));
      kname = "skl_map_vec";
    } else {
      grid = ceil_div(n, per_block);
      kname = "skl_map_sc";
    }
    launch(ctx, g, s->prog, kname, dim3((unsigned)grid), dim3(s->block), 0, args.data());
  };
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) {
    const Range r = core_range(in->units(), ctx->G, din, g);
    std::vector<Ready>& ch = chunks[(size_t)g];
    if (r.empty()) {
      ctx->set_device(g);
      for (const Ready& rd : ch) {  // nothing to compute here: just order the stream
        SKL_CUDA(cudaStreamWaitEvent(ctx->D(g).stream, rd.ev, 0));
        event_put(ctx, g, rd.ev);
      }
      continue;
    }
    ++ndev;
    size_t covered = 0;
    for (const Ready& rd : ch) {
      const size_t lo = std::max(rd.r.lo, r.lo), hi = std::min(rd.r.hi, r.hi);
      if (hi > lo) covered += hi - lo;
    }
    if (ch.empty() || covered != r.size()) {
      ctx->set_device(g);
      for (const Ready& rd : ch) {
        SKL_CUDA(cudaStreamWaitEvent(ctx->D(g).stream, rd.ev, 0));
        event_put(ctx, g, rd.ev);
      }
      launch_range(g, r);
      continue;
    }
    // pipelined: chunk k computes while chunk k+1 uploads; each output chunk
    // gets an event so that a download can stream it out while later chunks run
    for (const Ready& rd : ch) {
      const Range q{std::max(rd.r.lo, r.lo), std::min(rd.r.hi, r.hi)};
      ctx->set_device(g);
      SKL_CUDA(cudaStreamWaitEvent(ctx->D(g).stream, rd.ev, 0));
      event_put(ctx, g, rd.ev);
      if (q.empty()) continue;
      launch_range(g, q);
      if (o) {
        cudaEvent_t e = event_get(ctx, g);
        SKL_CUDA(cudaEventRecord(e, ctx->D(g).stream));
        o->parts[(size_t)g].ready.push_back(Ready{q, e});
      }
    }
  }
  if (o) mark_written(o);
  finish_extras(ctx, ea, ndev);
}

// ------------------------------------------------------------------ lazy fusion
void drop_lazy(Cont* c) {
  if (!c->lazy.s) return;
  for (Cont* in : {c->lazy.l, c->lazy.r})
    if (in) {
      auto& v = in->dependents;
      v.erase(std::remove(v.begin(), v.end(), c), v.end());
    }
  c->lazy = Lazy();
}

void materialize(Cont* c) {
  if (!c->lazy.s) return;
  const Lazy L = c->lazy;
  drop_lazy(c);
  Cont* o = c;
  c->dist = Dist();  // run_elementwise sets the output distribution
  // containers deferred on c want exactly the value computed now: keep them
  // deferred (prepare_output would otherwise materialise them first)
  std::vector<Cont*> deps;
  deps.swap(c->dependents);
  try {
    run_elementwise(L.s, L.l, L.r, &o, nullptr, 0);
  } catch (...) {
    c->dependents.swap(deps);
    throw;
  }
  c->dependents.swap(deps);
}

void materialize_dependents(Cont* c) {
  while (!c->dependents.empty()) materialize(c->dependents.back());
}

void run_map(Skel* s, Cont* in, Cont** out, const skl_arg* extra, int nextra) {
  if (s->kind != K_MAP) fail(SKL_ERR_INVALID_ARG, "not a Map skeleton");
  run_elementwise(s, in, nullptr, out, extra, nextra);
}
void run_zip(Skel* s, Cont* l, Cont* r, Cont** out, const skl_arg* extra, int nextra) {
  if (s->kind != K_ZIP) fail(SKL_ERR_INVALID_ARG, "not a Zip skeleton");
  if (!r) fail(SKL_ERR_INVALID_ARG, "zip needs two inputs");
  run_elementwise(s, l, r, out, extra, nextra);
}

// ------------------------------------------------------------------ Reduce
// What a device folds: the plain input, or (lazy fusion) the elements of a
// deferred Zip/Map computed from its inputs on the fly.
struct RedSrc {
  Program* prog;
  const char* kvec;
  const char* ksc;
  const void* p1;
  const void* p2;  // fused Zip: right input (Map: unused)
  bool vec_ok;
};

// One device's fold of n elements into `result` (device pointer).
static void reduce_on_device(Skel* s, int g, const RedSrc& src, size_t n, void* result) {
  Ctx* ctx = s->ctx;
  const size_t st = ctx->type(s->tin).size;
  const int nw = s->block / 32;
  const bool vec = (16 % st == 0) && src.vec_ok;
  const size_t rtile = 32 * (vec ? 16 / st : 1);
  const size_t ru = 4;
  // one wave of resident blocks (each warp owns a long segment: a second wave
  // would double the time)
  const char* kname = vec ? src.kvec : src.ksc;
  const size_t occ = (size_t)std::max(1, occupancy(ctx, g, src.prog, kname, s->block, 0));
  const size_t max_blocks = (size_t)ctx->D(g).sm_count * occ;
  size_t nblocks = std::min(max_blocks, std::max<size_t>(1, ceil_div(n, (size_t)nw * rtile * ru)));
  size_t wseg = ceil_div(ceil_div(n, nblocks * (size_t)nw), rtile) * rtile;
  nblocks = ceil_div(n, (size_t)nw * wseg);
  // scratch: [counter (16 B)] [partials]
  char* sc = (char*)scratch(s, s->scratch_red, g, 16 + max_blocks * std::max<size_t>(st, 8), true);
  void* counter = sc;
  void* partials = sc + 16;
  unsigned long long nn = n, ws = wseg;
  const void* p1 = src.p1;
  const void* p2 = src.p2;
  void* args1[] = {(void*)&p1, &nn, &ws, &partials, &counter, &result};
  void* args2[] = {(void*)&p1, (void*)&p2, &nn, &ws, &partials, &counter, &result};
  launch(ctx, g, src.prog, vec ? src.kvec : src.ksc, dim3((unsigned)nblocks), dim3(s->block), 0,
         src.p2 || std::strcmp(src.kvec, "skl_reduce_zip_vec") == 0 ? args2 : args1);
}

void run_combine(Skel* s, int g, const void* staging, size_t stride_elems, int nrep, void* dst,
                 size_t nelem) {
  if (!s || (s->kind != K_REDUCE && s->kind != K_SCAN)) fail(SKL_ERR_INVALID_ARG, "combine needs a Reduce skeleton");
  Ctx* ctx = s->ctx;
  unsigned long long stride = stride_elems, n = nelem;
  // 16-byte path: the element size divides 16, the replica stride is a whole
  // number of 16-byte words and both buffers are 16-byte aligned
  const size_t st = ctx->type(s->tin).size;
  int vec = 16 % st == 0 && st < 16 && (stride_elems * st) % 16 == 0 && aligned16(staging) && aligned16(dst);
  const size_t per = vec ? 16 / st : 1;
  const size_t grid = std::max<size_t>(1, std::min<size_t>(ceil_div(ceil_div(nelem, per), (size_t)s->block),
                                                           (size_t)ctx->D(g).sm_count * 8));
  void* args[] = {(void*)&staging, &stride, &nrep, &dst, &n, &vec};
  launch(ctx, g, s->prog, "skl_combine", dim3((unsigned)grid), dim3(s->block), 0, args);
}

// copy(+) -> block fused with its exchange (reduce.cuh skl_combine_peer): srcs
// are nrep <= 8 device pointers (this device's and its peers' replicas at the
// slice), dst this device's replica at the slice (may equal srcs[g]).
void run_combine_peer(Skel* s, int g, const void* const* srcs, int nrep, void* dst, size_t nelem) {
  if (!s || (s->kind != K_REDUCE && s->kind != K_SCAN)) fail(SKL_ERR_INVALID_ARG, "combine needs a Reduce skeleton");
  if (nrep < 1 || nrep > 8) fail(SKL_ERR_INVALID_ARG, "run_combine_peer: 1..8 replicas");
  Ctx* ctx = s->ctx;
  struct {
    const void* p[8];
  } sp{};
  const size_t st = ctx->type(s->tin).size;
  // 16-byte path when every source and the destination share one offset within
  // 16 bytes (a block slice that starts mid-word: its head is folded scalar)
  const uintptr_t mis = (uintptr_t)dst & 15u;
  int vec = 16 % st == 0 && st < 16 && mis % st == 0;
  for (int r = 0; r < nrep; ++r) {
    sp.p[r] = srcs[r];
    vec = vec && ((uintptr_t)srcs[r] & 15u) == mis;
  }
  int head = vec ? (int)(((16 - mis) & 15u) / st) : 0;
  unsigned long long n = nelem;
  const size_t per = vec ? 16 / st : 1;
  if (ceil_div(nelem, per) >= (1ull << 31)) fail(SKL_ERR_INVALID_ARG, "copy(+) combine: slice too large");
  // one pass: every thread folds s->cunr chunks (no grid-stride loop)
  const size_t grid = std::max<size_t>(1, ceil_div(ceil_div(nelem, per), (size_t)kCombineBlock * (size_t)s->cunr));
  void* args[] = {(void*)&sp, &nrep, &dst, &n, &vec, &head};
  launch(ctx, g, s->prog, "skl_combine_peer", dim3((unsigned)grid), dim3(kCombineBlock), 0, args);
}

// The same for logical devices sharing one GPU: one launch on device g over all
// n elements; bases[h] = replica h at unit 0, element e goes to replica
// e / chunk_elems.
void run_combine_all(Skel* s, int g, const void* const* bases, int nrep, size_t nelem, size_t chunk_elems) {
  if (!s || (s->kind != K_REDUCE && s->kind != K_SCAN)) fail(SKL_ERR_INVALID_ARG, "combine needs a Reduce skeleton");
  if (nrep < 1 || nrep > 8) fail(SKL_ERR_INVALID_ARG, "run_combine_all: 1..8 replicas");
  Ctx* ctx = s->ctx;
  struct {
    const void* p[8];
  } sp{};
  const size_t st = ctx->type(s->tin).size;
  // 16-byte loads whenever the replicas are 16-byte aligned; a chunk that
  // straddles two devices' slices is stored element by element
  int vec = 16 % st == 0 && st < 16;
  for (int r = 0; r < nrep; ++r) {
    sp.p[r] = bases[r];
    vec = vec && aligned16(bases[r]);
  }
  unsigned long long n = nelem, ch = chunk_elems;
  const size_t per = vec ? 16 / st : 1;
  if (ceil_div(nelem, per) >= (1ull << 31)) fail(SKL_ERR_INVALID_ARG, "copy(+) combine: container too large");
  const size_t grid = std::max<size_t>(1, ceil_div(ceil_div(nelem, per), (size_t)kCombineBlock * (size_t)s->cunr));
  void* args[] = {(void*)&sp, &nrep, &n, &ch, &vec};
  launch(ctx, g, s->prog, "skl_combine_all", dim3((unsigned)grid), dim3(kCombineBlock), 0, args);
}

// Fused program: the Zip/Map's and the Reduce's customising functions in one
// NVRTC program (each renamed by a macro, so both may be called "func"), the
// Reduce template reading through SklLoadZip.  nullptr if they do not compile
// together (then the Zip/Map is materialised instead).
static Program* fused_program(Skel* s, Skel* z) {
  auto it = s->fused.find(z);
  if (it != s->fused.end()) return it->second;
  Ctx* ctx = s->ctx;
  const size_t st = ctx->type(s->tin).size;
  const std::string zf = "skl_zf_" + z->entry, rf = "skl_rf_" + s->entry;
  std::string defs = defs_common(ctx, rf, s->block);
  defs += "#define SKL_T " + tname(ctx, s->tin) + "\n";
  defs += "#define SKL_RVEC " + std::to_string((16 % st == 0) ? 16 / st : 1) + "\n#define SKL_RU 4\n";
  defs += "#define SKL_FUSED 1\n#define SKL_ZL " + tname(ctx, z->tin) + "\n";
  defs += "#define SKL_ZR " + tname(ctx, z->kind == K_ZIP ? z->tin2 : z->tin) + "\n";
  defs += std::string("#define SKL_ZMAP ") + (z->kind == K_MAP ? "1" : "0") + "\n#define SKL_ZFUNC " + zf + "\n";
  const std::string body =
      "\n#define " + z->entry + " " + zf + "\n#line 1 \"user_source_zip\"\n" + z->user_src + "\n#undef " +
      z->entry + "\n#define " + s->entry + " " + rf + "\n#line 1 \"user_source_reduce\"\n" + s->user_src +
      "\n#undef " + s->entry + "\n#line 1 \"skeleton_template\"\n" + kernel_template("common.cuh") +
      kernel_template("op.cuh") + kernel_template("reduce.cuh");
  Program* p = nullptr;
  try {
    p = compile(ctx, defs + program_source(ctx, body), nullptr);
  } catch (const Error&) {
    p = nullptr;
  }
  s->fused[z] = p;
  return p;
}

void run_reduce(Skel* s, Cont* in, Cont** out) {
  if (s->kind != K_REDUCE) fail(SKL_ERR_INVALID_ARG, "not a Reduce skeleton");
  Ctx* ctx = s->ctx;
  if (in->elt != ctx->type(s->tin).size) fail(SKL_ERR_TYPE, "input type does not match the skeleton");
  if (in->rows * in->cols == 0) fail(SKL_ERR_EMPTY, "reduce of an empty container (A11)");
  // lazy fusion: fold a deferred Zip/Map straight from its inputs
  Lazy L = in->lazy;
  Program* fp = (L.s && ctx->lazy_fusion) ? fused_program(s, L.s) : nullptr;
  Dist din;
  if (fp) {
    din = L.d;
    ensure(L.l, L.l->dist.kind == DOVERLAP ? L.l->dist : din, false);
    if (L.r) {
      if (!(elementwise(L.r->dist) == din && L.r->dev_valid)) ensure(L.r, din, false);
      else ensure(L.r, L.r->dist, false);
    }
  } else {
    if (in->dist.kind == DCOPY && in->diverged && in->combine) ensure(in, Dist{DCOPY, 0}, false);
    din = elementwise(default_dist(in, Dist{DBLOCK, 0}));
    ensure(in, in->dist.kind == DOVERLAP ? in->dist : din, false);
  }
  Cont* o = output_for(ctx, out, s->tin, 1, 1, false);
  auto source = [&](int g, const Range& r) {
    if (fp) {
      const void* a = part_ptr(L.l, g, r.lo);
      const void* b = L.r ? part_ptr(L.r, g, r.lo) : nullptr;
      const bool eq = ctx->type(L.s->tin).size == in->elt &&
                      (!L.r || ctx->type(L.s->tin2).size == in->elt);
      return RedSrc{fp, "skl_reduce_zip_vec", "skl_reduce_zip_sc", a, b,
                    eq && aligned16(a) && (!b || aligned16(b))};
    }
    const void* a = part_ptr(in, g, r.lo);
    return RedSrc{s->prog, "skl_reduce_vec", "skl_reduce_sc", a, nullptr, aligned16(a)};
  };
  // participants, in device order: devices whose core holds elements.  A copy
  // input is reduced once per process (replicas are identical).
  std::vector<int> parts;
  for (int g = 0; g < ctx->G; ++g) {
    if (din.kind == DCOPY) {
      if (ctx->dist_mode ? g == ctx->first_local : g == 0) parts.push_back(g);
      continue;
    }
    if (!core_range(in->units(), ctx->G, din, g).empty()) parts.push_back(g);
  }
  // result distribution: single(first participant) in one process; copy across
  // processes so every rank's getValue() works (SPMD, A33).
  const bool cross = parts.size() > 1;
  Dist dout = ctx->dist_mode ? Dist{DCOPY, 0} : Dist{DSINGLE, parts[0]};
  if (!ctx->dist_mode && cross) dout = Dist{DSINGLE, 0};
  prepare_output(o, dout, 0);
  const size_t st = in->elt;
  if (!cross) {
    // one device computes everything
    for (int g : parts) {
      if (!ctx->is_local(g)) continue;
      const Range r = core_range(in->units(), ctx->G, din, g);
      reduce_on_device(s, g, source(g, r), r.size() * in->cols, part_ptr(o, g, 0));
    }
    mark_written(o);
    return;
  }
  // per-device partials (into slot p of a staging row), then gather + ordered fold
  const int P = (int)parts.size();
  std::map<int, void*> stage;  // device -> [P] staging
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g)
    stage[g] = scratch(s, s->scratch_stage, g, (size_t)P * std::max<size_t>(st, 8) + 64, false);
  std::vector<int> dsts;
  if (dout.kind == DSINGLE) dsts.push_back(dout.arg);
  else for (int g = 0; g < ctx->G; ++g) dsts.push_back(g);
  for (int i = 0; i < P; ++i) {
    const int g = parts[(size_t)i];
    if (!ctx->is_local(g)) continue;
    const Range r = core_range(in->units(), ctx->G, din, g);
    // partial lands in its own slot i on its own device
    reduce_on_device(s, g, source(g, r), r.size() * in->cols, (char*)stage[g] + (size_t)i * st);
  }
  // one process driving every device: the destination folds the partials
  // straight out of the participants' memory (peer loads), one kernel, no copy
  // (the same gate as the copy(+)->block fold: xfer_kernel=0 turns every peer kernel off)
  bool fused = ctx->combine_peer && ctx->xfer_kernel && !ctx->dist_mode && ctx->nlocal == ctx->G && P <= 8 &&
               dsts.size() == 1;
  for (int i = 0; fused && i < P; ++i) fused = ctx->peer_ok[(size_t)dsts[0]][(size_t)parts[(size_t)i]];
  if (fused) {
    std::vector<const void*> srcs((size_t)P);
    for (int i = 0; i < P; ++i) srcs[(size_t)i] = (char*)stage[parts[(size_t)i]] + (size_t)i * st;
    barrier_streams(ctx);  // every partial is written
    run_combine_peer(s, dsts[0], srcs.data(), P, part_ptr(o, dsts[0], 0), 1);
    barrier_streams(ctx);  // no device rewrites its partial slot while it is read
    mark_written(o);
    return;
  }
  std::vector<Transfer> tr;
  for (int dg : dsts)
    for (int i = 0; i < P; ++i)
      if (parts[(size_t)i] != dg) tr.push_back(Transfer{parts[(size_t)i], dg, 0, 0, 1, i});
  struct SPtr : PtrFn {
    std::map<int, void*>* stage;
    size_t st;
    void* src(const Transfer& t) override { return (char*)(*stage)[t.src] + (size_t)t.slot * st; }
    void* dst(const Transfer& t) override { return (char*)(*stage)[t.dst] + (size_t)t.slot * st; }
  } sp;
  sp.stage = &stage;
  sp.st = st;
  run_transfers(ctx, tr, st, sp);
  for (int dg : dsts)
    if (ctx->is_local(dg)) run_combine(s, dg, stage[dg], 1, P, part_ptr(o, dg, 0), 1);
  mark_written(o);
}

// ------------------------------------------------------------------ Scan
void run_scan(Skel* s, Cont* in, Cont** out) {
  if (s->kind != K_SCAN) fail(SKL_ERR_INVALID_ARG, "not a Scan skeleton");
  Ctx* ctx = s->ctx;
  if (in->elt != ctx->type(s->tin).size) fail(SKL_ERR_TYPE, "input type does not match the skeleton");
  if (in->rows * in->cols == 0) fail(SKL_ERR_EMPTY, "scan of an empty container");
  if (in->dist.kind == DCOPY && in->diverged && in->combine) ensure(in, Dist{DCOPY, 0}, false);
  const Dist din = elementwise(default_dist(in, Dist{DBLOCK, 0}));
  ensure(in, in->dist.kind == DOVERLAP ? in->dist : din, false);
  Cont* o = output_for(ctx, out, s->tin, in->rows, in->cols, in->matrix);
  if (o == in) fail(SKL_ERR_INVALID_ARG, "scan cannot run in place");
  prepare_output(o, din, 0);
  const size_t st = in->elt;
  const bool chunked = s->scan_ch > 0;
  const int items = chunked ? (int)((size_t)s->scan_ch * 16 / st) : 8;
  // participants with distinct data (block / single); copy scans whole on each device
  std::vector<int> parts;
  for (int g = 0; g < ctx->G; ++g)
    if (!core_range(in->units(), ctx->G, din, g).empty()) parts.push_back(g);
  const bool carry = din.kind == DBLOCK && parts.size() > 1;
  const int P = (int)parts.size();
  std::map<int, void*> totals;
  if (carry) {
    // pass 1: device totals (order-preserving reduce), all-gathered so device g
    // folds t_0 .. t_{g-1} as its carry-in
    for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g)
      totals[g] = scratch(s, s->scratch_stage, g, (size_t)P * std::max<size_t>(st, 8) + 64, false);
    for (int i = 0; i < P; ++i) {
      const int g = parts[(size_t)i];
      if (!ctx->is_local(g)) continue;
      const Range r = core_range(in->units(), ctx->G, din, g);
      {
        const void* a = part_ptr(in, g, r.lo);
        reduce_on_device(s, g, RedSrc{s->prog, "skl_reduce_vec", "skl_reduce_sc", a, nullptr, aligned16(a)},
                         r.size() * in->cols, (char*)totals[g] + (size_t)i * st);
      }
    }
    std::vector<Transfer> tr;
    for (int j = 0; j < P; ++j)
      for (int i = 0; i < j; ++i) tr.push_back(Transfer{parts[(size_t)i], parts[(size_t)j], 0, 0, 1, i});
    struct TPtr : PtrFn {
      std::map<int, void*>* t;
      size_t st;
      void* src(const Transfer& x) override { return (char*)(*t)[x.src] + (size_t)x.slot * st; }
      void* dst(const Transfer& x) override { return (char*)(*t)[x.dst] + (size_t)x.slot * st; }
    } tp;
    tp.t = &totals;
    tp.st = st;
    run_transfers(ctx, tr, st, tp);
  }
  for (int i = 0; i < P; ++i) {
    const int g = parts[(size_t)i];
    if (!ctx->is_local(g)) continue;
    const Range r = core_range(in->units(), ctx->G, din, g);
    const size_t n = r.size() * in->cols;
    const void* pin = part_ptr(in, g, r.lo);
    void* pout = part_ptr(o, g, r.lo);
    const bool vec = chunked && aligned16(pin) && aligned16(pout);
    // look-back unit: a chunk of scan_sub tiles (vector kernel) or one tile of 8 items
    // per thread (generic kernel)
    const size_t tile = (size_t)s->block * (size_t)(vec ? items : 8);
    const bool per_tile = s->scan_variant >= 2;  // one block per tile, tile look-back
    const size_t ntiles = ceil_div(n, vec && !per_tile ? tile * (size_t)s->scan_sub : tile);
    // status: [flags u32 x units] [aggs T x units] [incls T x units], 16-B aligned
    // packed status (elements <= 4 bytes): one u64 per tile holds value and flag
    // (status words are s->scan_fstride x 8 bytes apart: one L2 line per unit by default)
    const size_t fbytes = ceil_div(ntiles * 8 * (size_t)s->scan_fstride, 16) * 16,
                 tbytes = ceil_div(ntiles * st, 16) * 16;
    Scratch& sc = s->scratch_scan[g];
    const bool fresh = sc.bytes < fbytes + 2 * tbytes;
    char* base = (char*)scratch(s, s->scratch_scan, g, fbytes + 2 * tbytes, true);
    if (fresh) s->epoch[g] = 0;  // zeroed flags: every epoch >= 1 is new
    unsigned ep = ++s->epoch[g];
    if (ep >= (1u << 30)) {
      ctx->set_device(g);
      SKL_CUDA(cudaMemsetAsync(base, 0, fbytes, ctx->D(g).stream));
      ep = s->epoch[g] = 1;
    }
    void* flags = base;
    void* aggs = base + fbytes;
    void* incls = base + fbytes + tbytes;
    unsigned long long nn = n;
    const void* cptr = carry ? totals[g] : nullptr;
    int ncarry = carry ? i : 0;
    void* args[] = {(void*)&pin, &pout, &nn, &flags, &aggs, &incls, &ep, (void*)&cptr, &ncarry};
    if (vec && per_tile && (s->scan_variant == 6 || s->scan_variant == 7)) {
      // low-register per-tile kernel (tile in shared memory)
      const size_t smem = (size_t)s->block * (size_t)s->scan_ch * 16;
      launch(ctx, g, s->prog, "skl_scan_lr", dim3((unsigned)ntiles), dim3(s->block), smem, args);
    } else if (vec && per_tile && s->scan_variant >= 4) {
      // persistent 3-stage pipeline: one wave of resident blocks
      const size_t smem = 3 * (size_t)s->block * (size_t)s->scan_ch * 16;
      const int occ = std::max(1, occupancy(ctx, g, s->prog, "skl_scan_pipe", s->block, smem));
      const size_t grid = std::min(ntiles, (size_t)ctx->D(g).sm_count * (size_t)occ);
      launch(ctx, g, s->prog, "skl_scan_pipe", dim3((unsigned)grid), dim3(s->block), smem, args);
    } else if (vec && per_tile) {
      const size_t smem = (size_t)s->block * (size_t)s->scan_ch * 16;
      launch(ctx, g, s->prog, "skl_scan_pt", dim3((unsigned)ntiles), dim3(s->block), smem, args);
    } else if (vec) {
      // persistent grid (one wave of resident blocks), two shared-memory stages
      const size_t smem = 2 * (size_t)s->block * (size_t)s->scan_ch * 16;
      const int occ = std::max(1, occupancy(ctx, g, s->prog, "skl_scan_vec", s->block, smem));
      const size_t grid = std::min(ntiles, (size_t)ctx->D(g).sm_count * (size_t)occ);
      launch(ctx, g, s->prog, "skl_scan_vec", dim3((unsigned)grid), dim3(s->block), smem, args);
    } else {
      launch(ctx, g, s->prog, "skl_scan_sc", dim3((unsigned)ntiles), dim3(s->block), 0, args);
    }
  }
  mark_written(o);
}

// ------------------------------------------------------------------ MapOverlap
// Fused halo push: with every device of a block-distributed
// output in this process, device g's kernel also stores its first / last d
// units into the halo units of devices g-1 / g+1 (peer memory over NVLink, or
// the same GPU for logical devices), so a following overlap(d) read moves no
// data.  Taken only when every core holds >= d units (each halo unit then has
// exactly one producer, the adjacent device) and peer stores are possible.
static bool plan_halo_push(Ctx* ctx, Cont* o, size_t d, std::vector<void*>& up, std::vector<void*>& down) {
  const int G = ctx->G;
  if (!ctx->halo_push || G < 2 || d == 0 || o->dist.kind != DBLOCK) return false;
  if (ctx->ipc) {
    // one process per GPU over NVLink: the neighbours' output parts, exchanged
    // (collective: every rank takes the same decision from the same values)
    up.assign((size_t)G, nullptr);
    down.assign((size_t)G, nullptr);
    const int me = ctx->first_local;
    const Range want = need_range(o->units(), G, Dist{DOVERLAP, (int)d}, me);
    const Part& p = o->parts[(size_t)me];
    const bool ok = p.ptr && p.buf.contains(want);
    const auto all = ipc_exchange(ctx, {(uint64_t)(uintptr_t)p.ptr, (uint64_t)p.buf.lo, ok ? 1u : 0u});
    for (int g = 0; g < G; ++g)
      if (core_range(o->units(), G, o->dist, g).size() < d || all[(size_t)g].at(2) == 0) return false;
    const Range r = core_range(o->units(), G, o->dist, me);
    const size_t ub = o->unit_bytes();
    if (me > 0)
      up[(size_t)me] = (char*)ipc_translate(ctx, me - 1, all[(size_t)me - 1][0]) + (r.lo - all[(size_t)me - 1][1]) * ub;
    if (me + 1 < G)
      down[(size_t)me] =
          (char*)ipc_translate(ctx, me + 1, all[(size_t)me + 1][0]) + (r.hi - d - all[(size_t)me + 1][1]) * ub;
    return true;
  }
  if (ctx->dist_mode || ctx->nlocal != G) return false;
  up.assign((size_t)G, nullptr);
  down.assign((size_t)G, nullptr);
  for (int g = 0; g < G; ++g) {
    const Range r = core_range(o->units(), G, o->dist, g);
    if (r.size() < d) return false;
    const Range want = need_range(o->units(), G, Dist{DOVERLAP, (int)d}, g);
    const Part& p = o->parts[(size_t)g];
    if (!p.ptr || !p.buf.contains(want)) return false;
    if (g > 0 && !ctx->peer_ok[(size_t)g][(size_t)g - 1]) return false;
    if (g + 1 < G && !ctx->peer_ok[(size_t)g][(size_t)g + 1]) return false;
  }
  for (int g = 0; g < G; ++g) {
    const Range r = core_range(o->units(), G, o->dist, g);
    if (g > 0) up[(size_t)g] = part_ptr(o, g - 1, r.lo);
    if (g + 1 < G) down[(size_t)g] = part_ptr(o, g + 1, r.hi - d);
  }
  return true;
}

// TMA descriptor of a device's input part for skl_mo2d_t / skl_mo2d_ws: a 2-D
// tiled map over rows x columns (row pitch C * elt bytes, a multiple of 16),
// box = the staged window (pitch x srows elements).  The row is described in
// 2^ushift-byte units: the widest of 8/4/2/1 bytes that divides the window's
// width and offsets in bytes (every window starts at a multiple of 16 bytes:
// tile widths and the halo width A are 16-byte multiples), so a byte image's
// 544-byte window is 68 units, inside the 256-unit box limit.  Returns false
// when TMA cannot describe it (box wider than 256 units or taller than 256
// rows, no driver entry point): the caller uses skl_mo2d.
static bool encode_tile_map(SklTensorMap* tm, const void* base, size_t elt, size_t C, size_t rows, size_t pitch,
                            size_t srows, int* ushift) {
  static PFN_cuTensorMapEncodeTiled_v12000 enc = nullptr;
  static bool tried = false;
  if (!tried) {
    tried = true;
    cudaDriverEntryPointQueryResult q;
    void* fn = nullptr;
    if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &fn, cudaEnableDefault, &q) == cudaSuccess &&
        q == cudaDriverEntryPointSuccess)
      enc = (PFN_cuTensorMapEncodeTiled_v12000)fn;
    else
      (void)cudaGetLastError();
  }
  if (!enc) return false;
  const size_t wb = pitch * elt;  // window width in bytes (a multiple of 16)
  const size_t unit = wb % 8 == 0 ? 8 : wb % 4 == 0 ? 4 : wb % 2 == 0 ? 2 : 1;
  if ((C * elt) % unit != 0) return false;
  const size_t units = wb / unit, cu = C * elt / unit;
  if (units > 256 || srows > 256 || rows == 0 || rows >= (1ull << 31) || cu >= (1ull << 31)) return false;
  const CUtensorMapDataType dt = unit == 8 ? CU_TENSOR_MAP_DATA_TYPE_UINT64
                                 : unit == 4 ? CU_TENSOR_MAP_DATA_TYPE_UINT32
                                 : unit == 2 ? CU_TENSOR_MAP_DATA_TYPE_UINT16
                                             : CU_TENSOR_MAP_DATA_TYPE_UINT8;
  const cuuint64_t dims[2] = {(cuuint64_t)cu, (cuuint64_t)rows};
  const cuuint64_t strides[1] = {(cuuint64_t)(C * elt)};
  const cuuint32_t box[2] = {(cuuint32_t)units, (cuuint32_t)srows};
  const cuuint32_t estr[2] = {1, 1};
  const CUresult r = enc((CUtensorMap*)tm, dt, 2, const_cast<void*>(base), dims, strides, box, estr,
                         CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE,
                         CU_TENSOR_MAP_L2_PROMOTION_L2_128B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  if (r != CUDA_SUCCESS) return false;
  *ushift = unit == 8 ? 3 : unit == 4 ? 2 : unit == 2 ? 1 : 0;
  return true;
}

void run_mapoverlap(Skel* s, Cont* in, Cont** out) {
  if (s->kind != K_MAPOVERLAP) fail(SKL_ERR_INVALID_ARG, "not a MapOverlap skeleton");
  Ctx* ctx = s->ctx;
  if (in->elt != ctx->type(s->tin).size) fail(SKL_ERR_TYPE, "input type does not match the skeleton");
  const int d = s->d;
  // A4/A6: the input must be overlap(d' >= d) (or copy / single, computed whole)
  Dist din = in->dist;
  if (din.kind == DNONE || din.kind == DBLOCK || (din.kind == DOVERLAP && din.arg < d))
    din = Dist{DOVERLAP, d};
  ensure(in, din, true);
  const Dist dout = (din.kind == DOVERLAP) ? Dist{DBLOCK, 0} : din;
  Cont* o = output_for(ctx, out, s->tout, in->rows, in->cols, in->matrix);
  if (o == in) fail(SKL_ERR_INVALID_ARG, "MapOverlap cannot run in place");
  if (in->rows >= (1ull << 31) || in->cols >= (1ull << 31))
    fail(SKL_ERR_INVALID_ARG, "MapOverlap: rows and columns must be < 2^31");
  prepare_output(o, dout, dout.kind == DBLOCK ? (size_t)d : 0);
  const size_t si = in->elt, so = o->elt;
  std::vector<void*> push_up, push_down;
  const bool push = plan_halo_push(ctx, o, (size_t)d, push_up, push_down);
  long hd = push ? (long)d : 0;
  // the pushes overwrite halo units the neighbours may still be reading
  if (push) {
    if (ctx->ipc) ipc_barrier(ctx);
    else barrier_streams(ctx);
  }
  auto push_ptrs = [&](int g, void** pu, void** pd) {
    *pu = push ? push_up[(size_t)g] : nullptr;
    *pd = push ? push_down[(size_t)g] : nullptr;
    if (*pu) ctx->pushed += (long long)((size_t)d * o->unit_bytes());
    if (*pd) ctx->pushed += (long long)((size_t)d * o->unit_bytes());
  };
  if (in->matrix) {
    for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) {
      const Range r = core_range(in->units(), ctx->G, dout, g);
      if (r.empty()) continue;
      Part& pi = in->parts[(size_t)g];
      Part& po = o->parts[(size_t)g];
      const void* pin = pi.ptr;
      void* pout = po.ptr;
      long in_row0 = (long)pi.buf.lo, in_rows = (long)pi.buf.size(), out_row0 = (long)po.buf.lo;
      long R = (long)in->rows, C = (long)in->cols, rb = (long)r.lo, re = (long)r.hi;
      const int cw = s->mo_tw / 32;
      void *pu, *pd;
      push_ptrs(g, &pu, &pd);
      const size_t ow = (size_t)cw * so;
      int vec_ok = ((size_t)C * si) % 16 == 0 && aligned16(pin) && ((size_t)C * so) % ow == 0 &&
                   (uintptr_t)pout % ow == 0 && (uintptr_t)pu % ow == 0 && (uintptr_t)pd % ow == 0;
      void* args[] = {(void*)&pin, &in_row0, &in_rows, &pout, &out_row0, &R, &C, &rb, &re,
                      s->neutral.data(), &vec_ok, &pu, &pd, &hd};
      const dim3 grid((unsigned)ceil_div((size_t)C, (size_t)s->mo_tw),
                      (unsigned)ceil_div(r.size(), (size_t)s->mo_th));
      SklTensorMap tm;
      int ushift = 0;
      // fix: TMA-staged border tiles need patching unless the boundary value is zero
      int fix = s->boundary == 1 ? 1 : 0;
      for (unsigned char b : s->neutral) fix |= b != 0;
      const bool tma = (ctx->mo_ws || (ctx->mo_tma && !ctx->mo_persist)) && vec_ok &&
                       encode_tile_map(&tm, pin, si, (size_t)C, (size_t)in_rows, (size_t)s->mo_pitch,
                                       (size_t)(s->mo_th + 2 * s->d), &ushift);
      if (tma && !ctx->mo_ws) {
        // s->mo_kt vertically stacked tiles per block, each staged by one TMA copy
        // issued up front (skl_mo2d_t); the count is chosen at creation
        const int kt = s->mo_kt;
        const size_t ts = ((size_t)(s->mo_th + 2 * s->d) * (size_t)s->mo_pitch * si + 127) / 128 * 128;
        const size_t smem = kt > 1 ? (size_t)kt * ts + 128 : 0;
        const dim3 tgrid(grid.x, (unsigned)ceil_div(r.size(), (size_t)s->mo_th * (size_t)kt));
        void* targs[] = {(void*)&tm, &pout, &in_row0, &out_row0, &R, &C, &rb, &re, s->neutral.data(), &vec_ok,
                         &pu, &pd, &hd, &fix, &ushift};
        launch(ctx, g, s->prog, "skl_mo2d_t", tgrid, dim3(s->block), smem, targs);
        ctx->n_tma++;
      } else if (tma) {
        // TMA producer warp + consumer warps over a ring of staged tiles
        const size_t tile_bytes = (size_t)(s->mo_th + 2 * s->d) * (size_t)s->mo_pitch * si;
        const int nst = ctx->mo_ws_stages;
        const size_t smem = (size_t)nst * ((tile_bytes + 127) / 128 * 128) + 128;
        int tiles_x = (int)grid.x, ntiles = (int)(grid.x * grid.y);
        const int nthr = s->block + 32;
        const int occ = std::max(1, occupancy(ctx, g, s->prog, "skl_mo2d_ws", nthr, smem));
        const size_t pgrid = std::min((size_t)ntiles, (size_t)ctx->D(g).sm_count * (size_t)occ);
        void* wargs[] = {(void*)&tm, &pout, &in_row0, &out_row0, &R, &C, &rb, &re, s->neutral.data(), &vec_ok,
                         &pu, &pd, &hd, &tiles_x, &ntiles, (void*)&nst, &fix, &ushift};
        launch(ctx, g, s->prog, "skl_mo2d_ws", dim3((unsigned)pgrid), dim3((unsigned)nthr), smem, wargs);
        ctx->n_tma++;
      } else if (ctx->mo_persist) {
        // resident blocks walk the tiles with two staging buffers (load of tile
        // k+1 overlaps f on tile k)
        const size_t tile_bytes = (size_t)(s->mo_th + 2 * s->d) * (size_t)s->mo_pitch * si;
        const size_t smem = 2 * tile_bytes;
        int tiles_x = (int)grid.x, ntiles = (int)(grid.x * grid.y);
        const int occ = std::max(1, occupancy(ctx, g, s->prog, "skl_mo2d_p", s->block, smem));
        const size_t pgrid = std::min((size_t)ntiles, (size_t)ctx->D(g).sm_count * (size_t)occ);
        void* pargs[] = {(void*)&pin, &in_row0, &in_rows, &pout, &out_row0, &R, &C, &rb, &re,
                         s->neutral.data(), &vec_ok, &pu, &pd, &hd, &tiles_x, &ntiles};
        launch(ctx, g, s->prog, "skl_mo2d_p", dim3((unsigned)pgrid), dim3(s->block), smem, pargs);
      } else {
        launch(ctx, g, s->prog, "skl_mo2d", grid, dim3(s->block), 0, args);
      }
    }
  } else {
    // vector form: compile the 1-D variant once
    if (!s->prog1d) {
      const size_t epc = 16 / si;
      const int A = (int)(ceil_div((size_t)d, epc) * epc);
      const int cw = 4, tw = s->block * cw;
      std::string defs = defs_common(ctx, s->entry, s->block);
      defs += "#define SKL_TIN " + tname(ctx, s->tin) + "\n#define SKL_TOUT " + tname(ctx, s->tout) + "\n";
      defs += "#define SKL_D " + std::to_string(d) + "\n#define SKL_BOUNDARY " + std::to_string(s->boundary) + "\n";
      defs += "#define SKL_A " + std::to_string(A) + "\n#define SKL_PITCH 0\n";
      defs += "#define SKL_TW " + std::to_string(tw) + "\n#define SKL_TH 1\n#define SKL_CW " +
              std::to_string(cw) + "\n#define SKL_RH 1\n#define SKL_MO1D 1\n#define SKL_OUTB " +
              std::to_string((size_t)cw * ctx->type(s->tout).size) + "\n#define SKL_SO " +
              std::to_string(ctx->type(s->tout).size) + "\n";
      const std::string user = "\n#line 1 \"user_source\"\n" + s->user_src + "\n#line 1 \"skeleton_template\"\n";
      s->prog1d = compile(ctx, defs + program_source(ctx, user + kernel_template("common.cuh") +
                                                                   kernel_template("mapoverlap.cuh")),
                                nullptr);
      s->mo_1d = true;
    }
    const int tw = s->block * 4;
    for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) {
      const Range r = core_range(in->units(), ctx->G, dout, g);
      if (r.empty()) continue;
      Part& pi = in->parts[(size_t)g];
      Part& po = o->parts[(size_t)g];
      const void* pin = pi.ptr;
      void* pout = po.ptr;
      long in_lo = (long)pi.buf.lo, in_n = (long)pi.buf.size(), out_lo = (long)po.buf.lo;
      long N = (long)in->rows, unused = 0, rb = (long)r.lo, re = (long)r.hi;
      int vec_ok = aligned16(pin);
      void *pu, *pd;
      push_ptrs(g, &pu, &pd);
      void* args[] = {(void*)&pin, &in_lo, &in_n, &pout, &out_lo, &N, &unused, &rb, &re,
                      s->neutral.data(), &vec_ok, &pu, &pd, &hd};
      launch(ctx, g, s->prog1d, "skl_mo1d", dim3((unsigned)ceil_div(r.size(), (size_t)tw)),
             dim3(s->block), 0, args);
    }
  }
  mark_written(o);
  if (push) {
    o->halo_ready = (size_t)d;
    // the neighbours' next reads of their halos wait for the pushes
    if (ctx->ipc) ipc_barrier(ctx);
    else barrier_streams(ctx);
  }
  if (ctx->debug_bounds) check_debug_flag(ctx);
}

void check_debug_flag(Ctx* ctx) {
  extern bool read_and_clear_bounds_flags(Ctx*);
  if (read_and_clear_bounds_flags(ctx))
    fail(SKL_ERR_OUT_OF_RANGE, "get() accessed an element beyond the overlap range d (P:L362-368)");
}

}  // namespace skl
