// allpairs.cpp — the Allpairs skeleton.
//
// allpairs(+)(A, B) = C with C[i][j] = A_i (+) B_j over the rows of A (n x d)
// and B (m x d).  Distribution ("block(A) x copy(B)"): A keeps
// its distribution (default block rows, A6), B becomes copy (every device needs
// all of it), C rows follow A's.  No exchange is needed.
#include <algorithm>

#include "skl_internal.h"

namespace skl {

namespace {
size_t cdiv(size_t a, size_t b) { return (a + b - 1) / b; }
}  // namespace

Skel* allpairs_create(Ctx* ctx, const char* src, const char* entry, const char* rsrc,
                      const char* rentry, int tin, int tout) {
  if (!src) fail(SKL_ERR_INVALID_ARG, "customising function source is NULL");
  const size_t si = ctx->type(tin).size, so = ctx->type(tout).size;
  if (si == 0 || so == 0) fail(SKL_ERR_TYPE, "Allpairs needs non-void types");
  auto s = std::make_unique<Skel>();
  s->ctx = ctx;
  s->kind = K_ALLPAIRS;
  s->user_src = src;
  s->entry = (entry && *entry) ? std::string(entry) : detect_entry(s->user_src);
  s->tin = tin;
  s->tout = tout;
  s->block = 256;
  s->ap_zr = rsrc != nullptr;
  std::string defs = "#define SKL_BLOCK 256\n#define SKL_DEBUG_BOUNDS 0\n";
  defs += std::string("#define SKL_AP_FAST ") + (si == 4 ? "1" : "0") + "\n";
  if (ctx->ap_bk) defs += "#define SKL_AP_BK " + std::to_string(ctx->ap_bk) + "\n";
  defs += "#define SKL_TIN " + ctx->type(tin).name + "\n#define SKL_TOUT " + ctx->type(tout).name + "\n";
  std::string body;
  if (s->ap_zr) {
    const std::string rs = rsrc;
    const std::string re = (rentry && *rentry) ? std::string(rentry) : detect_entry(rs);
    const std::string zf = "skl_zf_" + s->entry, rf = "skl_rf_" + re;
    defs += "#define SKL_AP_ZR 1\n#define SKL_ZFUNC " + zf + "\n#define SKL_RFUNC " + rf + "\n";
    // both functions may carry the same name ("func"): rename each by macro
    body = "\n#define " + s->entry + " " + zf + "\n#line 1 \"user_source_zip\"\n" + s->user_src +
           "\n#undef " + s->entry + "\n#define " + re + " " + rf + "\n#line 1 \"user_source_reduce\"\n" + rs +
           "\n#undef " + re + "\n#line 1 \"skeleton_template\"\n";
    s->user_src += "\n" + rs;  // kept for introspection
  } else {
    defs += "#define SKL_AP_ZR 0\n#define SKL_FUNC " + s->entry + "\n";
    body = "\n#line 1 \"user_source\"\n" + s->user_src + "\n#line 1 \"skeleton_template\"\n";
  }
  body += kernel_template("common.cuh") + kernel_template("allpairs.cuh");
  s->prog = compile(ctx, defs + program_source(ctx, body), nullptr);
  Skel* raw = s.release();
  ctx->skels.insert(raw);
  return raw;
}

void run_allpairs(Skel* s, Cont* a, Cont* b, Cont** out) {
  if (s->kind != K_ALLPAIRS) fail(SKL_ERR_INVALID_ARG, "not an Allpairs skeleton");
  Ctx* ctx = s->ctx;
  const size_t si = ctx->type(s->tin).size;
  if (a->elt != si || b->elt != si) fail(SKL_ERR_TYPE, "Allpairs inputs do not match the skeleton's type");
  if (!a->matrix || !b->matrix) fail(SKL_ERR_TYPE, "Allpairs takes two matrices (rows are the entities)");
  if (a->cols != b->cols) fail(SKL_ERR_SIZE_MISMATCH, "Allpairs: A and B rows differ in length d");
  const size_t n = a->rows, m = b->rows, d = a->cols;
  if (d == 0) fail(SKL_ERR_EMPTY, "Allpairs of zero-length rows");
  Dist din = a->dist.kind == DNONE ? Dist{DBLOCK, 0} : a->dist;
  if (din.kind == DOVERLAP) din = Dist{DBLOCK, 0};
  ensure(a, a->dist.kind == DOVERLAP ? a->dist : din, false);
  ensure(b, Dist{DCOPY, 0}, false);
  Cont* c = *out;
  if (c) {
    if (c->type != s->tout || c->rows != n || c->cols != m)
      fail(SKL_ERR_SIZE_MISMATCH, "Allpairs output must be an n x m matrix of the output type");
  } else {
    c = cont_create(ctx, s->tout, n, m, true);
    *out = c;
  }
  prepare_output(c, din, 0);
  for (int g = ctx->first_local; g < ctx->first_local + ctx->nlocal; ++g) {
    const Range r = core_range(n, ctx->G, din, g);
    if (r.empty()) continue;
    const void* pa = part_ptr(a, g, r.lo);
    const void* pb = part_ptr(b, g, 0);
    void* pc = part_ptr(c, g, r.lo);
    long nn = (long)r.size(), mm = (long)m, dd = (long)d;
    if (s->ap_zr) {
      void* args[] = {(void*)&pa, (void*)&pb, &pc, &nn, &mm, &dd};
      const bool fast = si == 4 && d % 4 == 0 && ((uintptr_t)pa % 16) == 0 && ((uintptr_t)pb % 16) == 0 &&
                        ctx->ap_fast;
      if (fast) {
        // 128 x 128 tiles (2 blocks/SM) or 128 x 64 (3 blocks/SM): the one whose
        // tile count fills the last wave better (option ap_tile forces 8 / 4)
        const size_t sms = (size_t)ctx->D(g).sm_count, rows = cdiv(r.size(), 128);
        const size_t t8 = cdiv(m, 128) * rows, t4 = cdiv(m, 64) * rows;
        auto eff = [](size_t t, size_t slots) { return (double)t / (double)(cdiv(t, slots) * slots); };
        // 128 x 64 measured ~17 % slower per FLOP (4096^3: 5.42 vs 4.98 ms): only for poor wave fill
        bool narrow = eff(t4, 3 * sms) * 0.82 > eff(t8, 2 * sms);
        if (ctx->ap_tile == 8) narrow = false;
        if (ctx->ap_tile == 4) narrow = true;
        // hybrid: whole waves of 128 x 128 tiles, the partial last wave as
        // 128 x 64 halves (when they fit one wave of 2 blocks per SM)
        // shared memory: two stages of (128 + tile columns) rows x (bk + 4) elements
        const size_t bk = ctx->ap_bk ? (size_t)ctx->ap_bk : 16;
        const size_t sm8 = 2 * (128 + 128) * (bk + 4) * si, sm4 = 2 * (128 + 64) * (bk + 4) * si;
        const size_t slots = 2 * sms, rem = t8 % slots;
        const bool hybrid = (ctx->ap_tile == 0 || ctx->ap_tile == 2) && ctx->ap_hybrid && t8 > slots &&
                            rem != 0 && 2 * rem <= slots;
        if (hybrid || ctx->ap_tile == 2) {
          long nwide = (long)(t8 - rem), tiles_x = (long)cdiv(m, 128);
          void* hargs[] = {(void*)&pa, (void*)&pb, &pc, &nn, &mm, &dd, &nwide, &tiles_x};
          launch(ctx, g, s->prog, "skl_ap_zrh", dim3((unsigned)(t8 + rem)), dim3(256), sm8, hargs);
        } else if (narrow)
          launch(ctx, g, s->prog, "skl_ap_zr4", dim3((unsigned)cdiv(m, 64), (unsigned)rows), dim3(256), sm4, args);
        else
          launch(ctx, g, s->prog, "skl_ap_zr8", dim3((unsigned)cdiv(m, 128), (unsigned)rows), dim3(256), sm8, args);
      } else {
        launch(ctx, g, s->prog, "skl_ap_zr", dim3((unsigned)cdiv(m, 64), (unsigned)cdiv(r.size(), 64)),
               dim3(256), 0, args);
      }
    } else {
      const size_t smem = 32 * (d + 1) * si;
      int use_smem = smem <= 96 * 1024;
      void* args[] = {(void*)&pa, (void*)&pb, &pc, &nn, &mm, &dd, &use_smem};
      launch(ctx, g, s->prog, "skl_ap_gen", dim3((unsigned)cdiv(m, 16), (unsigned)cdiv(r.size(), 16)),
             dim3(256), use_smem ? smem : 0, args);
    }
  }
  mark_written(c);
}

}  // namespace skl
