"""CPU-only tests of the C-ABI library (no GPU here): libskl.so loads without a
CUDA driver, exports every symbol include/skl.h declares, NVRTC compiles every
skeleton template for sm_100a (offline context), compile errors
come back as SKL_ERR_COMPILE with the log, and the host-side distribution
planner matches the oracle's partition rule."""
import os
import re
import subprocess
import tempfile

import numpy as np
import pytest

import oracle as O
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import build as B
from paper_conf_pact_steuwerg13_b200 import skl as S

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def lib():
    B.build()
    return S.lib()


def header_symbols():
    txt = open(os.path.join(ROOT, "include", "skl.h")).read()
    return sorted(set(re.findall(r"\b(skl_[a-z0-9_]+)\s*\(", txt)) - {"skl_arg"})


def test_library_exports_every_declared_symbol(lib):
    so = os.path.join(ROOT, "paper_conf_pact_steuwerg13_b200", "libskl.so")
    out = subprocess.run(["nm", "-D", "--defined-only", so], capture_output=True, text=True).stdout
    exported = set(re.findall(r" T (skl_[a-z0-9_]+)", out))
    declared = header_symbols()
    assert len(declared) >= 40
    missing = [s for s in declared if s not in exported]
    assert not missing, missing


def test_library_has_no_link_time_cuda_driver_dependency(lib):
    so = os.path.join(ROOT, "paper_conf_pact_steuwerg13_b200", "libskl.so")
    ldd = subprocess.run(["ldd", so], capture_output=True, text=True).stdout
    assert "libcuda.so" not in ldd and "not found" not in ldd


def test_init_without_gpu_fails_loudly(lib):
    # no GPU in this container: the product path must refuse, not fall back
    import torch
    if torch.cuda.is_available():
        pytest.skip("GPU present")
    with pytest.raises(S.SklError) as e:
        S.Context()
    assert e.value.name == "CUDA"


@pytest.fixture(scope="module")
def offline(lib):
    ctx = S.Context.offline()
    yield ctx
    ctx.finalize()


def _sass(skel) -> str:
    with tempfile.NamedTemporaryFile(suffix=".cubin", delete=False) as f:
        f.write(skel.cubin())
        p = f.name
    try:
        return subprocess.run(["cuobjdump", "-sass", p], capture_output=True, text=True).stdout
    finally:
        os.unlink(p)


def test_offline_compiles_every_skeleton_for_sm100a(offline):
    ctx = offline
    aff = ctx.struct_type("Aff", A.AFFINE_DECL, 8, 4)
    ev = ctx.struct_type("Event", A.EVENT_DECL, A.EVENT_SIZE, 4)
    sks = [
        S.Map(ctx, A.NEG, S.F32, S.F32), S.Map(ctx, A.mandelbrot(1000), S.F32X2, S.U32),
        S.Map(ctx, A.INV_U8, S.U8, S.U8), S.Map(ctx, A.AFFINE_I32, S.I32, S.I32),
        S.Zip(ctx, A.MULT, S.F32, S.F32, S.F32), S.Zip(ctx, A.SUB_I32, S.I32, S.I32, S.I32),
        S.Reduce(ctx, A.SUM, S.F32), S.Reduce(ctx, A.AFFINE_COMPOSE, aff), S.Reduce(ctx, A.ADD_F64, S.F64),
        S.Scan(ctx, A.ADD, S.F32), S.Scan(ctx, A.ADD_I32, S.I32), S.Scan(ctx, A.AFFINE_COMPOSE, aff),
        S.MapOverlap(ctx, A.SOBEL, S.U8, S.U8, 1, S.NEUTRAL, 0),
        S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0),
        S.MapOverlap(ctx, A.BOX3, S.F32, S.F32, 1, S.NEUTRAL, 0.0),
        S.Map(ctx, A.lmosem_map(150), ev, S.VOID, extra=[S.F32 | S.PTR, S.F32 | S.PTR]),
    ]
    for sk in sks:
        cub = sk.cubin()
        assert len(cub) > 1000 and cub[:4] == b"\x7fELF"
    # the sm_100a kernels exist in the cubin with the skeleton entry points
    sass = _sass(sks[0])
    assert "skl_map_vec" in sass and "sm_100a" in sass
    assert "LDG.E.ENL2.128" in sass or "LDG.E.128" in sass or ".128" in sass


def test_paper_strings_compile_with_entry_detection(offline):
    # the function name differs per string
    for src in (A.NEG, A.ADD, A.SUM, A.MULT):
        assert "SKL_FUNC" in S.Map(offline, src, S.F32, S.F32).source() if src == A.NEG else True
    s = S.Zip(offline, "// helper first\nfloat twice(float v){return 2.0f*v;}\n" + A.MULT,
              S.F32, S.F32, S.F32).source()
    assert "#define SKL_FUNC mult" in s


def test_fmad_disabled_in_generated_code(offline):
    sass = _sass(S.Map(offline, A.SQP1, S.F32, S.F32))
    assert "FFMA" not in sass and "FMUL" in sass and "FADD" in sass


def test_compile_error_reports_log(offline):
    with pytest.raises(S.SklError) as e:
        S.Map(offline, "float f(float x){ return undefined_name; }", S.F32, S.F32)
    assert e.value.name == "COMPILE" and "undefined_name" in str(e.value)


def test_type_errors(offline):
    with pytest.raises(S.SklError):
        S.MapOverlap(offline, A.IDENT2D, S.F32, S.F32, -1)
    ev = offline.struct_type("Ev3", "struct Ev3 { float a, b, c; };", 12, 4)
    with pytest.raises(S.SklError) as e:
        S.MapOverlap(offline, "float f(const Ev3* p){ return get(p,0,0).a; }", ev, S.F32, 1)
    assert e.value.name == "TYPE"


@pytest.mark.parametrize("units", [0, 1, 7, 100, 3072, 8193])
@pytest.mark.parametrize("G", [1, 2, 3, 4, 8])
def test_planner_matches_oracle_partition(lib, units, G):
    for g in range(G):
        assert S.plan_range(units, G, S.BLOCK, 0, g, False) == O.block_range(units, G, g)
        assert S.plan_range(units, G, S.OVERLAP, 2, g, True) == O.overlap_range(units, G, g, 2)
        assert S.plan_range(units, G, S.OVERLAP, 2, g, False) == O.block_range(units, G, g)
        assert S.plan_range(units, G, S.COPY, 0, g, False) == (0, units)
        assert S.plan_range(units, G, S.SINGLE, G - 1, g, False) == ((0, units) if g == G - 1 else (0, 0))


def _simulate(units, G, fk, fa, tk, ta):
    """apply the planned transfers to per-device dicts {unit: value}; check the
    target layout holds exactly the right units with the right values."""
    have = []
    for g in range(G):
        lo, hi = S.plan_range(units, G, fk, fa, g, fk == S.OVERLAP)
        have.append({u: u for u in range(lo, hi)})
    new = [dict() for _ in range(G)]
    for g in range(G):  # local reuse
        lo, hi = S.plan_range(units, G, tk, ta, g, tk == S.OVERLAP)
        for u in range(lo, hi):
            if u in have[g]:
                new[g][u] = have[g][u]
    for src, su, dst, du, n in S.plan_transfers(units, G, fk, fa, tk, ta):
        assert src != dst
        for k in range(n):
            assert su + k in have[src]          # the source really holds it
            assert du + k not in new[dst]       # never moved twice / overwritten
            new[dst][du + k] = have[src][su + k]
    for g in range(G):
        lo, hi = S.plan_range(units, G, tk, ta, g, tk == S.OVERLAP)
        assert new[g] == {u: u for u in range(lo, hi)}


DISTS = [(S.SINGLE, 0), (S.SINGLE, 1), (S.COPY, 0), (S.BLOCK, 0), (S.OVERLAP, 1), (S.OVERLAP, 3)]


@pytest.mark.parametrize("fk,fa", DISTS)
@pytest.mark.parametrize("tk,ta", DISTS)
@pytest.mark.parametrize("units,G", [(10, 2), (17, 4), (5, 8), (64, 3)])
def test_planned_redistribution_is_exact(lib, fk, fa, tk, ta, units, G):
    if (fk == S.SINGLE and fa >= G) or (tk == S.SINGLE and ta >= G):
        pytest.skip()
    _simulate(units, G, fk, fa, tk, ta)


# ------------------------------------------------------------------ static get() bounds
def test_static_get_bounds(offline):
    c = offline
    # Listing 1.2 (counted loops), Listing 1.5 (literals), the 5x5 Gaussian: proven
    assert S.MapOverlap(c, A.BOX3, S.F32, S.F32, 1).bounds_proven
    assert S.MapOverlap(c, A.SOBEL, S.U8, S.U8, 1).bounds_proven
    assert S.MapOverlap(c, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST).bounds_proven
    assert S.MapOverlap(c, A.BOX1D, S.F32, S.F32, 1).bounds_proven
    # provable violations are rejected at creation, before any kernel runs
    for src, d in (("float f(const float* p){ return get(p, 2, 0); }", 1),
                   ("float f(const float* p){ return get(p, 0, -3); }", 2),
                   ("float f(float* m){ float s=0; for (int i = -2; i <= 2; ++i) s += get(m, i, 0); return s; }", 1),
                   ("float f(float* m){ float s=0; for (int j = 0; j <= 3; j++) s += get(m, 0, j); return s; }", 2)):
        with pytest.raises(S.SklError) as e:
            S.MapOverlap(c, src, S.F32, S.F32, d)
        assert e.value.name == "OUT_OF_RANGE"
    # the same loops within d are proven; a runtime offset is not provable
    assert S.MapOverlap(c, "float f(float* m){ float s=0; for (int j = 0; j < 3; j++) s += get(m, 0, j); return s; }",
                        S.F32, S.F32, 2).bounds_proven
    assert not S.MapOverlap(c, "float f(const float* p){ int k = 1; return get(p, k, 0); }",
                            S.F32, S.F32, 1).bounds_proven
    # comments do not count
    assert S.MapOverlap(c, "float f(const float* p){ /* get(p, 9, 9) */ return get(p, 1, 1); }",
                        S.F32, S.F32, 1).bounds_proven


def test_disk_cache_and_env_defaults(tmp_path, monkeypatch):
    """SKL_CACHE_DIR: a second context loads the cubin from disk instead of
    running NVRTC; SKL_BLOCK_THREADS / SKL_DEBUG_BOUNDS set context defaults
    (SURVEY §5 config).  Offline contexts: no GPU needed."""
    monkeypatch.setenv("SKL_CACHE_DIR", str(tmp_path))
    src = "float twice(float x){ return x + x; }"
    c1 = S.Context.offline()
    S.Map(c1, src, S.F32, S.F32)
    assert c1.counter("compiles") == 1 and c1.counter("disk_cache_hits") == 0
    c1.finalize()
    assert len(list(tmp_path.glob("skl_*.cubin"))) == 1
    c2 = S.Context.offline()
    m = S.Map(c2, src, S.F32, S.F32)
    assert c2.counter("compiles") == 0 and c2.counter("disk_cache_hits") == 1
    assert len(m.cubin()) > 0
    c2.finalize()
    monkeypatch.setenv("SKL_BLOCK_THREADS", "128")
    c3 = S.Context.offline()
    assert "#define SKL_BLOCK 128" in S.Map(c3, src, S.F32, S.F32).source()
    c3.finalize()


def test_map_over_a_loop_defaults_to_one_element_per_lane(offline):
    """map_auto: a customising function with a loop (Mandelbrot's A22 escape
    loop) compiles the interleaved kernel with one element per lane; a
    straight-line function keeps the 16-byte chunks; comments and strings
    mentioning loops do not count; map_auto 0 turns it off"""
    def ilj(src, tin=S.F32, tout=S.F32):
        s = S.Map(offline, src, tin, tout).source()
        return int(s.split("#define SKL_ILJ ")[1].split()[0])
    assert ilj(A.mandelbrot(100), S.F32X2, S.U32) == 1
    assert ilj("float f(float x){ float s = 0.0f; for (int k = 0; k < 3; ++k) s = s + x; return s; }") == 1
    assert ilj(A.NEG) > 1
    assert ilj("float f(float x){ /* for while */ return x + 1.0f; } // do") > 1
    offline.set_option("map_auto", 0)
    try:
        assert ilj(A.mandelbrot(100), S.F32X2, S.U32) > 1
    finally:
        offline.set_option("map_auto", 1)
