"""Small cases of every kernel for compute-sanitizer, each checked
against the oracle so a sanitizer run is also a parity run:

  compute-sanitizer --tool memcheck  --error-exitcode 3 python tools/sanitize_cases.py
  compute-sanitizer --tool racecheck --error-exitcode 3 python tools/sanitize_cases.py
  compute-sanitizer --tool synccheck --error-exitcode 3 python tools/sanitize_cases.py
"""
import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tests"))

import oracle as O  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import apps as A  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import inputs as I  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import skl as S  # noqa: E402
from paper_conf_pact_steuwerg13_b200.lmosem import ListModeOSEM  # noqa: E402


def rel(a, b):
    a, b = np.asarray(a, np.float64), np.asarray(b, np.float64)
    return float(np.linalg.norm(a - b) / max(np.linalg.norm(b), 1e-300))


def one_device(opts):
    ctx = S.Context(1)
    for k, v in opts.items():
        ctx.set_option(k, v)
    n = 70001
    x = I.uniform_f32(1, n) - np.float32(0.5)
    y = I.uniform_f32(2, n)
    vx, vy = S.Vector.from_numpy(ctx, x), S.Vector.from_numpy(ctx, y)
    assert np.array_equal(S.Map(ctx, A.SQP1, S.F32, S.F32)(vx).to_numpy(), O.map_(O.OM_SQP1_F32, x))
    assert np.array_equal(S.Zip(ctx, A.ADD, S.F32, S.F32, S.F32)(vx, vy).to_numpy(), O.zip_(O.OZ_ADD_F32, x, y))
    u = I.uniform_int(3, n, 0, 255, np.int64).astype(np.uint8)
    assert np.array_equal(S.Map(ctx, A.INV_U8, S.U8, S.U8)(S.Vector.from_numpy(ctx, u)).to_numpy(),
                          O.map_(O.OM_INV_U8, u))
    red = S.Reduce(ctx, A.SUM, S.F32)
    ref = O.reduce_(O.OP_ADD_F32, x)
    assert abs(float(red(vx).scalar()) - ref) <= 1e-5 * max(1.0, abs(ref))
    d = float(red(S.Zip(ctx, A.MULT, S.F32, S.F32, S.F32)(vx, vy)).scalar())   # fused
    dref = O.reduce_(O.OP_ADD_F32, O.zip_(O.OZ_MULT_F32, x, y))
    assert abs(d - dref) <= 1e-5 * max(1.0, abs(dref))
    xi = I.uniform_int(4, n, -1000, 1000)
    sc = S.Scan(ctx, A.ADD_I32, S.I32)
    assert np.array_equal(sc(S.Vector.from_numpy(ctx, xi)).to_numpy(), O.scan(O.OP_ADD_I32, xi))
    aff = ctx.struct_type("Aff", A.AFFINE_DECL, 8, 4)
    p = I.uniform_int(5, 2 * 5003, 0, 2**32 - 1, np.uint64).astype(np.uint32).reshape(5003, 2)
    got = S.Scan(ctx, A.AFFINE_COMPOSE, aff)(S.Vector(ctx, aff, 5003).copy_in(p)).to_numpy(np.uint32)
    assert np.array_equal(got.reshape(5003, 2), O.scan(O.OP_AFFINE_U32, p))
    img8 = I.image_u8(5, 70, 133)
    sob = S.MapOverlap(ctx, A.SOBEL, S.U8, S.U8, 1, S.NEUTRAL, 0)
    assert np.array_equal(sob(S.Matrix.from_numpy(ctx, img8)).to_numpy(),
                          O.mapoverlap2d(O.OS_SOBEL, img8, 1, O.OB_NEUTRAL, 0))
    imgf = I.image_f32(6, 150, 270)
    gau = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
    assert np.array_equal(gau(S.Matrix.from_numpy(ctx, imgf)).to_numpy(),
                          O.mapoverlap2d(O.OS_GAUSS5, imgf, 2, O.OB_NEAREST, 0.0))
    v1 = I.uniform_f32(7, 9001)
    box1 = S.MapOverlap(ctx, A.BOX1D, S.F32, S.F32, 1, S.NEAREST, 0.0)
    assert np.array_equal(box1(S.Vector.from_numpy(ctx, v1)).to_numpy(),
                          O.mapoverlap1d(O.OS_BOX3, v1, 1, O.OB_NEAREST, 0.0))
    a = I.uniform_f32(8, 130 * 36).reshape(130, 36)
    b = I.uniform_f32(9, 70 * 36).reshape(70, 36)
    for src, red_src, fn in ((A.MULT, A.ADD, O.AP_DOT), (A.MANHATTAN_ROWS, None, O.AP_MANHATTAN)):
        ap = S.Allpairs(ctx, src, S.F32, S.F32, reduce=red_src) if red_src else S.Allpairs(ctx, src, S.F32, S.F32)
        assert np.array_equal(ap(S.Matrix.from_numpy(ctx, a), S.Matrix.from_numpy(ctx, b)).to_numpy(),
                              O.allpairs(fn, a, b))
    grid = I.mandel_grid(24, 32)
    m = S.Map(ctx, A.mandelbrot_unrolled(1000, 8), S.F32X2, S.U32)
    assert np.array_equal(m(S.Matrix(ctx, S.F32X2, 24, 32).copy_in(grid)).to_numpy(), O.mandelbrot(grid, 1000)[0])
    ctx.finalize()


def logical_devices(G):
    ctx = S.Context(G, devices=[0] * G)
    x = I.uniform_f32(11, 10007)
    v = S.Vector.from_numpy(ctx, x).set_distribution(S.BLOCK)
    v.set_distribution(S.COPY)
    v.set_distribution(S.SINGLE, G - 1)
    v.set_distribution(S.OVERLAP, 3)
    v.set_distribution(S.BLOCK)
    assert np.array_equal(v.to_numpy(), x)
    sc = S.Scan(ctx, A.ADD, S.F32)
    assert rel(sc(v).to_numpy(), O.scan(O.OP_ADD_F32, x)) <= 1e-5
    imgf = I.image_f32(12, 61, 40)
    gau = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
    g2 = gau(gau(S.Matrix.from_numpy(ctx, imgf)))       # fused halo push between the two
    r1 = O.mapoverlap2d(O.OS_GAUSS5, imgf, 2, O.OB_NEAREST, 0.0)
    assert np.array_equal(g2.to_numpy(), O.mapoverlap2d(O.OS_GAUSS5, r1, 2, O.OB_NEAREST, 0.0))
    N, nev = 8, 3000
    osem = ListModeOSEM(ctx, N)
    ev = I.lmosem_events(13, nev, N)
    f0 = np.ones(N ** 3, np.float32)
    osem.load_events(ev, 2)
    osem.set_image(f0)
    osem.iterate(1)
    f = f0
    for lo, hi in ListModeOSEM.subset_bounds(nev, 2):
        f = O.lmosem(ev[lo:hi], N, f)[1].astype(np.float32)
    assert rel(osem.image(), f) <= 1e-4
    osem.destroy()
    # copy(+) -> block: one-launch fused fold (1), per-device fused kernels (2), staged (0)
    addf = S.Reduce(ctx, A.ADD, S.F32)
    idx = S.Vector.from_numpy(ctx, np.arange(5003, dtype=np.int32) % 4099).set_distribution(S.BLOCK)
    touch = S.Map(ctx, "void touch(int i, float* c) { atomicAdd(&c[i], 1.0f); }", S.I32, S.VOID,
                  extra=[S.F32 | S.PTR])
    want = np.bincount(np.arange(5003) % 4099, minlength=4099).astype(np.float32)
    for peer in (1, 2, 0):
        ctx.set_option("combine_peer", peer)
        cv = S.Vector(ctx, S.F32, 4099).set_distribution(S.COPY, 0, addf)
        cv.fill(0.0)
        touch(idx, (cv, S.WRITE))
        cv.set_distribution(S.BLOCK)
        assert np.array_equal(cv.to_numpy(), want)
    ctx.set_option("combine_peer", 1)
    ctx.finalize()


def tma_and_hybrid(G):
    """TMA / warp-specialised MapOverlap (mbarrier ring, border patching, parts
    with halo rows on G logical devices, fused halo push) and the hybrid Allpairs
    launch (every tile split)"""
    ctx = S.Context(G, devices=[0] * G)
    ctx.set_option("mo_ws", 1)
    ctx.set_option("mo_ws_stages", 2)
    ctx.set_option("mo_cw", 4)
    ctx.set_option("ap_tile", 2)
    n0 = ctx.counter("tma_launches")
    img8 = I.image_u8(5, 70, 144)
    sob = S.MapOverlap(ctx, A.SOBEL, S.U8, S.U8, 1, S.NEUTRAL, 0)
    assert np.array_equal(sob(S.Matrix.from_numpy(ctx, img8)).to_numpy(),
                          O.mapoverlap2d(O.OS_SOBEL, img8, 1, O.OB_NEUTRAL, 0))
    imgf = I.image_f32(6, 150, 272)
    gau = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
    g2 = gau(gau(S.Matrix.from_numpy(ctx, imgf)))
    r1 = O.mapoverlap2d(O.OS_GAUSS5, imgf, 2, O.OB_NEAREST, 0.0)
    assert np.array_equal(g2.to_numpy(), O.mapoverlap2d(O.OS_GAUSS5, r1, 2, O.OB_NEAREST, 0.0))
    assert ctx.counter("tma_launches") - n0 == 3 * G
    a = I.uniform_f32(8, 130 * 36).reshape(130, 36)
    b = I.uniform_f32(9, 200 * 36).reshape(200, 36)
    ap = S.Allpairs(ctx, A.MULT, S.F32, S.F32, reduce=A.ADD)
    assert np.array_equal(ap(S.Matrix.from_numpy(ctx, a).set_distribution(S.BLOCK),
                             S.Matrix.from_numpy(ctx, b)).to_numpy(), O.allpairs(O.AP_DOT, a, b))
    ctx.finalize()


def tma_tile_cases(G):
    """the default TMA tile kernel (skl_mo2d_t, 1 and 2 tiles per block, border
    patching, parts with halo rows, fused halo push) on G logical devices, both
    Sobel forms, and the one-pass copy(+) fold on slices that start mid-word"""
    for kt in (1, 2):
        ctx = S.Context(G, devices=[0] * G)
        ctx.set_option("mo_kt", kt)
        n0 = ctx.counter("tma_launches")
        img8 = I.image_u8(5, 70, 144)
        for src in (A.SOBEL, A.SOBEL_TUNED):
            sob = S.MapOverlap(ctx, src, S.U8, S.U8, 1, S.NEUTRAL, 0)
            s1 = sob(sob(S.Matrix.from_numpy(ctx, img8)))
            r8 = O.mapoverlap2d(O.OS_SOBEL, O.mapoverlap2d(O.OS_SOBEL, img8, 1, O.OB_NEUTRAL, 0), 1, O.OB_NEUTRAL, 0)
            assert np.array_equal(s1.to_numpy(), r8)
        # the tuned Sobel in the bench's 8 x 8 register block
        for k, v in (("mo_rh", 8), ("mo_cw", 8)):
            ctx.set_option(k, v)
        sob = S.MapOverlap(ctx, A.SOBEL_TUNED, S.U8, S.U8, 1, S.NEUTRAL, 0)
        assert np.array_equal(sob(sob(S.Matrix.from_numpy(ctx, img8))).to_numpy(), r8)
        for k in ("mo_rh", "mo_cw"):
            ctx.set_option(k, 0)
        imgf = I.image_f32(6, 150, 272)
        ctx.set_option("block_threads", 128)
        gau = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
        g2 = gau(gau(S.Matrix.from_numpy(ctx, imgf)))
        r1 = O.mapoverlap2d(O.OS_GAUSS5, imgf, 2, O.OB_NEAREST, 0.0)
        assert np.array_equal(g2.to_numpy(), O.mapoverlap2d(O.OS_GAUSS5, r1, 2, O.OB_NEAREST, 0.0))
        assert ctx.counter("tma_launches") - n0 == 8 * G
        n = 3001
        addf = S.Reduce(ctx, A.ADD, S.F32)
        cv = S.Vector(ctx, S.F32, n).set_distribution(S.COPY, 0, addf).fill(0.0)
        idx = S.Vector.from_numpy(ctx, np.arange(n, dtype=np.int32)).set_distribution(S.BLOCK)
        touch = S.Map(ctx, "void touch(int i, float* c) { c[i] = 1.0f + (float)(i % 5); }", S.I32, S.VOID,
                      extra=[S.F32 | S.PTR])
        touch(idx, (cv, S.WRITE))
        cv.set_distribution(S.BLOCK)
        assert np.array_equal(cv.to_numpy(), (1.0 + np.arange(n) % 5).astype(np.float32))
        ctx.finalize()


def graph_cases(G):
    """an iterated Gaussian on G logical devices (one stream each) recorded as ONE
    multi-device CUDA graph and replayed, halos pushed inside the graph; and a
    Map over a function with a loop (the interleaved one-element-per-lane default)"""
    import torch
    ctx = S.Context(G, devices=[0] * G)
    streams = [torch.cuda.Stream() for _ in range(G)]
    for g, st in enumerate(streams):
        ctx.set_stream(g, st.cuda_stream)
    gau = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
    img = I.image_f32(6, 97, 70)
    a = S.Matrix.from_numpy(ctx, img)
    b = S.Matrix(ctx, S.F32, 97, 70)
    t = S.Matrix(ctx, S.F32, 97, 70)

    def it():
        gau(a, out=b)
        gau(b, out=t)

    it()
    gr = ctx.capture(it)
    t.fill(0.0)
    gr.launch()
    gr.launch()
    ref = O.mapoverlap2d(O.OS_GAUSS5, O.mapoverlap2d(O.OS_GAUSS5, img, 2, O.OB_NEAREST, 0.0), 2, O.OB_NEAREST, 0.0)
    assert np.array_equal(t.to_numpy(), ref)
    gr.destroy()
    grid = I.mandel_grid(24, 40)
    m = S.Map(ctx, A.mandelbrot(200), S.F32X2, S.U32)
    x = S.Matrix(ctx, S.F32X2, 24, 40).set_distribution(S.BLOCK).copy_in(np.ascontiguousarray(grid))
    got = m(x).to_numpy(np.uint32).reshape(24, 40)
    assert np.array_equal(got, O.mandelbrot(grid, 200)[0])
    ctx.finalize()


if __name__ == "__main__":
    graph_cases(3)
    tma_tile_cases(1)
    tma_tile_cases(3)
    one_device({})
    one_device({"scan_variant": 3, "map_interleave": 1, "block_threads": 128})
    logical_devices(3)
    tma_and_hybrid(1)
    tma_and_hybrid(2)
    print("sanitize cases ok", flush=True)
