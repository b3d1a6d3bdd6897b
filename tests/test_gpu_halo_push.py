"""Fused halo push: on G devices in one process, a MapOverlap
whose output is block-distributed stores its border rows straight into the
neighbours' halo rows, so an iterated stencil (the paper's overlap use,
P:L214-222) needs no separate exchange between iterations.

Checked against the oracle applied T times, bit-exact, with and without the
push; the counters prove that the pushed run moved no device-to-device bytes
after the first iteration and that the fallback (cores smaller than d) still
exchanges halos by copies."""
import numpy as np
import pytest

import oracle as O
from gpu_util import require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu

T = 4


@pytest.fixture(scope="module", params=[2, 3, 4])
def ctx(request):
    require_gpu()
    c = S.Context(request.param, devices=[0] * request.param)
    yield c
    c.set_option("halo_push", 1)
    c.finalize()


def _oracle_iter(x, T, stencil, d, boundary):
    r = x
    for _ in range(T):
        r = O.mapoverlap2d(stencil, r, d, boundary, 0.0)
    return r


def _iterate(ctx, sk, x, T):
    """ping-pong between two output containers (the second iteration on writes
    into a container a neighbour device read as input one step earlier)"""
    m = S.Matrix.from_numpy(ctx, x)
    a = sk(m)
    b = S.Matrix(ctx, S.F32, x.shape[0], x.shape[1])
    p2p0, push0 = ctx.counter("p2p_bytes"), ctx.counter("halo_push_bytes")
    src, dst = a, b
    for _ in range(T - 1):
        sk(src, out=dst)
        src, dst = dst, src
    return src, ctx.counter("p2p_bytes") - p2p0, ctx.counter("halo_push_bytes") - push0


@pytest.mark.parametrize("shape", [(64, 200), (301, 257), (8, 33), (17, 16)])
def test_iterated_gauss_pushed(ctx, shape):
    G = ctx.ndev
    gau = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
    x = I.image_f32(I.SEED_GAUSS, *shape)
    want = _oracle_iter(x, T, O.OS_GAUSS5, 2, O.OB_NEAREST)
    ctx.set_option("halo_push", 1)
    got, p2p, pushed = _iterate(ctx, gau, x, T)
    assert np.array_equal(got.to_numpy(), want)
    assert got.distribution()[0] == S.BLOCK
    if shape[0] >= 2 * G:  # every core >= d = 2 rows: the push is taken
        assert p2p == 0
        # (T-1) launches per device, 2 neighbours for inner devices
        assert pushed == (T - 1) * 2 * (G - 1) * 2 * shape[1] * 4
    ctx.set_option("halo_push", 0)
    got0, p2p0, pushed0 = _iterate(ctx, gau, x, T)
    ctx.set_option("halo_push", 1)
    assert np.array_equal(got0.to_numpy(), want)
    assert pushed0 == 0 and p2p0 > 0


def test_small_cores_fall_back(ctx):
    """rows < d * G: some cores are shorter than the halo; exchange by copies"""
    G = ctx.ndev
    gau = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
    x = I.image_f32(I.SEED_GAUSS + 1, 2 * G - 1, 40)
    got, p2p, pushed = _iterate(ctx, gau, x, T)
    assert np.array_equal(got.to_numpy(), _oracle_iter(x, T, O.OS_GAUSS5, 2, O.OB_NEAREST))
    assert pushed == 0


def test_sobel_then_box(ctx):
    """u8 push (Sobel, d=1), then a different skeleton reads the pushed halos"""
    sob = S.MapOverlap(ctx, A.SOBEL, S.U8, S.U8, 1, S.NEUTRAL, 0)
    x = I.image_u8(I.SEED_SOBEL, 130, 96)
    s1 = sob(S.Matrix.from_numpy(ctx, x))
    p2p0 = ctx.counter("p2p_bytes")
    s2 = sob(s1)
    assert ctx.counter("p2p_bytes") == p2p0
    r1 = O.mapoverlap2d(O.OS_SOBEL, x, 1, O.OB_NEUTRAL, 0)
    assert np.array_equal(s2.to_numpy(), O.mapoverlap2d(O.OS_SOBEL, r1, 1, O.OB_NEUTRAL, 0))


def test_wider_overlap_needs_exchange(ctx):
    """halos pushed for d=1 do not satisfy an overlap(2) read: copies are used"""
    box = S.MapOverlap(ctx, A.BOX3, S.F32, S.F32, 1, S.NEAREST, 0.0)
    gau = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
    x = I.image_f32(I.SEED_GAUSS + 2, 96, 64)
    b = box(S.Matrix.from_numpy(ctx, x))
    p2p0 = ctx.counter("p2p_bytes")
    g = gau(b)
    assert ctx.counter("p2p_bytes") > p2p0
    r1 = O.mapoverlap2d(O.OS_BOX3, x, 1, O.OB_NEAREST, 0.0)
    assert np.array_equal(g.to_numpy(), O.mapoverlap2d(O.OS_GAUSS5, r1, 2, O.OB_NEAREST, 0.0))


def test_write_invalidates_pushed_halos(ctx):
    """a Map that rewrites the pushed container invalidates its halos"""
    box = S.MapOverlap(ctx, A.BOX3, S.F32, S.F32, 1, S.NEAREST, 0.0)
    neg = S.Map(ctx, A.NEG, S.F32, S.F32)
    x = I.image_f32(I.SEED_GAUSS + 3, 64, 48)
    b = box(S.Matrix.from_numpy(ctx, x))
    neg(b, out=b)  # in place: b's halos are stale now
    c = box(b)
    r1 = -O.mapoverlap2d(O.OS_BOX3, x, 1, O.OB_NEAREST, 0.0)
    assert np.array_equal(c.to_numpy(), O.mapoverlap2d(O.OS_BOX3, r1, 1, O.OB_NEAREST, 0.0))


def test_vector_pushed(ctx):
    box1 = S.MapOverlap(ctx, A.BOX1D, S.F32, S.F32, 1, S.NEAREST, 0.0)
    v = I.uniform_f32(91, 10007)
    a = box1(S.Vector.from_numpy(ctx, v))
    p2p0, push0 = ctx.counter("p2p_bytes"), ctx.counter("halo_push_bytes")
    b = box1(a)
    assert ctx.counter("p2p_bytes") == p2p0
    assert ctx.counter("halo_push_bytes") - push0 == 2 * (ctx.ndev - 1) * 4
    r1 = O.mapoverlap1d(O.OS_BOX3, v, 1, O.OB_NEAREST, 0.0)
    assert np.array_equal(b.to_numpy(), O.mapoverlap1d(O.OS_BOX3, r1, 1, O.OB_NEAREST, 0.0))


@pytest.mark.parametrize("push", [1, 0])
@pytest.mark.parametrize("G", [2, 3])
def test_multi_device_graph_replays_iterated_stencil(G, push):
    """three Gaussian iterations on G logical devices recorded as ONE CUDA graph
    (the capture forks into every device stream) and replayed: bit-exact
    against the oracle, with the halos pushed by the stencil or refreshed by
    copies inside the graph; the graph reads the containers at launch time"""
    require_gpu()
    c = S.Context(G, devices=[0] * G)
    try:
        c.set_option("halo_push", push)
        gau = S.MapOverlap(c, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
        img = I.image_f32(I.SEED_GAUSS + 3, 301, 203)
        a = S.Matrix.from_numpy(c, img)
        b = S.Matrix(c, S.F32, 301, 203)
        t = S.Matrix(c, S.F32, 301, 203)

        def it():
            gau(a, out=b)
            gau(b, out=t)
            gau(t, out=b)

        it()                                   # compiles, allocates, plans
        g = c.capture(it)
        ref = img
        for _ in range(3):
            ref = O.mapoverlap2d(O.OS_GAUSS5, ref, 2, O.OB_NEAREST, 0.0)
        for _ in range(2):
            b.fill(0.0)
            t.fill(0.0)
            g.launch()
            assert np.array_equal(b.to_numpy(), ref)
        img2 = I.image_f32(I.SEED_GAUSS + 4, 301, 203)
        a.copy_in(img2)
        g.launch()
        ref2 = img2
        for _ in range(3):
            ref2 = O.mapoverlap2d(O.OS_GAUSS5, ref2, 2, O.OB_NEAREST, 0.0)
        assert np.array_equal(b.to_numpy(), ref2)
        g.destroy()
    finally:
        c.finalize()
