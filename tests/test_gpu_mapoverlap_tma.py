"""GPU parity tests for the TMA-staged one-tile-per-block 2-D MapOverlap kernel
(skl_mo2d_t, option mo_tma, the default where a tensor map describes the part;
DESIGN.md 6.3): one cp.async.bulk.tensor copy stages a block's window, cells
outside the matrix are zero-filled by the copy engine and patched for NEAREST
and non-zero NEUTRAL (A20).  Bit-exact against the oracle at sizes
spanning several tiles with ragged edges, every boundary mode, byte and float
images, logical multi-device runs with the fused halo push; the per-thread
cp.async kernel (mo_tma=0) gives the same results.  Also the tuned Sobel user
function (apps.SOBEL_TUNED): full images in every register-block geometry and
its square-root step for every m."""
import re

import numpy as np
import pytest

import oracle as O
from gpu_util import require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu

SHAPES_F32 = [(1, 4), (3, 16), (37, 52), (65, 132), (200, 300), (513, 1000)]
SHAPES_U8 = [(1, 16), (3, 32), (37, 48), (65, 144), (200, 304), (513, 1008), (70, 1040)]


def tma_ctx(ndev=1, **opts):
    require_gpu()
    c = S.Context(ndev, devices=[0] * ndev)
    for k, v in opts.items():
        c.set_option(k, v)
    return c


@pytest.mark.parametrize("shape", SHAPES_F32)
@pytest.mark.parametrize("tma,kt", [(1, 2), (1, 1), (1, 4), (0, 2)])
def test_tma_f32_modes(shape, tma, kt):
    c = tma_ctx(mo_tma=tma, mo_kt=kt, block_threads=128)
    try:
        x = I.image_f32(I.SEED_GAUSS, *shape)
        m = S.Matrix.from_numpy(c, x)
        before = c.counter("tma_launches")
        for src, kind, d, bnd, nv in ((A.gaussian5(), O.OS_GAUSS5, 2, S.NEAREST, 0.0),
                                      (A.gaussian5(), O.OS_GAUSS5, 2, S.NEUTRAL, 0.0),
                                      (A.BOX3, O.OS_BOX3, 1, S.NEAREST, 0.0),
                                      (A.SHIFTX, O.OS_SHIFT_X, 1, S.NEUTRAL, 7.0),
                                      (A.SHIFTY, O.OS_SHIFT_Y, 1, S.NEAREST, 0.0)):
            mo = S.MapOverlap(c, src, S.F32, S.F32, d, bnd, nv)
            got = mo(m).to_numpy()
            ref = O.mapoverlap2d(kind, x, d, O.OB_NEAREST if bnd == S.NEAREST else O.OB_NEUTRAL, nv)
            assert np.array_equal(got, ref), (src, shape)
        # rows of 16-byte multiples go through TMA when it is on
        assert c.counter("tma_launches") - before == (5 if tma and (shape[1] * 4) % 16 == 0 else 0)
    finally:
        c.finalize()


@pytest.mark.parametrize("shape", SHAPES_U8)
@pytest.mark.parametrize("rh,tma,kt", [(0, 1, 2), (2, 1, 1), (4, 1, 3), (0, 0, 2)])
def test_tma_u8(shape, rh, tma, kt):
    c = tma_ctx(mo_rh=rh, mo_tma=tma, mo_kt=kt) if rh else tma_ctx(mo_tma=tma, mo_kt=kt)
    try:
        x = I.image_u8(I.SEED_SOBEL, *shape)
        m = S.Matrix.from_numpy(c, x)
        before = c.counter("tma_launches")
        for src in (A.SOBEL, A.SOBEL_TUNED):
            sob = S.MapOverlap(c, src, S.U8, S.U8, 1, S.NEUTRAL, 0)
            assert np.array_equal(sob(m).to_numpy(), O.mapoverlap2d(O.OS_SOBEL, x, 1, O.OB_NEUTRAL, 0)), src
        sx = S.MapOverlap(c, A.SHIFTX_U8, S.U8, S.U8, 1, S.NEAREST, 0)
        assert np.array_equal(sx(m).to_numpy(), O.mapoverlap2d(O.OS_SHIFT_X, x, 1, O.OB_NEAREST, 0))
        idn = S.MapOverlap(c, A.IDENT2D_U8, S.U8, S.U8, 1, S.NEUTRAL, 0)
        assert np.array_equal(idn(m).to_numpy(), x)
        assert c.counter("tma_launches") - before == (4 if tma else 0)
    finally:
        c.finalize()


@pytest.mark.parametrize("ndev", [2, 3])
@pytest.mark.parametrize("dt", ["f32", "u8"])
@pytest.mark.parametrize("tma", [1, 0])
def test_tma_overlap_distribution_and_halo_push(ndev, dt, tma):
    """parts with halo rows (the map starts at the part's first row), iterated
    stencils whose halos are pushed by the kernel into the neighbours"""
    c = tma_ctx(ndev, mo_tma=tma)
    try:
        if dt == "f32":
            x = I.image_f32(I.SEED_GAUSS, 301, 260)
            st = S.MapOverlap(c, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
            f = lambda r: O.mapoverlap2d(O.OS_GAUSS5, r, 2, O.OB_NEAREST, 0.0)  # noqa: E731
        else:
            x = I.image_u8(I.SEED_SOBEL, 301, 272)
            st = S.MapOverlap(c, A.SOBEL_TUNED, S.U8, S.U8, 1, S.NEUTRAL, 0)
            f = lambda r: O.mapoverlap2d(O.OS_SOBEL, r, 1, O.OB_NEUTRAL, 0)  # noqa: E731
        a = S.Matrix.from_numpy(c, x)
        b = st(a)
        t = st(b)
        b2 = st(t)
        ref = x
        for _ in range(3):
            ref = f(ref)
        assert np.array_equal(b2.to_numpy(), ref)
        assert c.counter("tma_launches") >= (3 * ndev if tma else 0)
        assert c.counter("halo_push_bytes") > 0
    finally:
        c.finalize()


def test_sobel_tuned_root_step_every_m():
    """the square-root step of apps.SOBEL_TUNED, cut out of the user function's
    own text (the bias added to m as the function adds it) and run as a Map over m = 0 .. 2^21 - 1 (h^2 + v^2 <= 2,080,800 <
    2^21), against numpy's correctly rounded fp32 root: min(255, (int)sqrtf(m))"""
    c = tma_ctx()
    try:
        src = A.SOBEL_TUNED
        last = "  return (uchar)__float_as_int(t);\n"
        body = src[src.index("  float k"):src.index(last) + len(last)]
        assert "sqrt.approx" in body and "add.rm" in body
        # the function's m carries the 2^23 exponent bias (added as the v*v
        # multiply-add's addend); here it is added to the plain m
        assert "int m = h * h + (v * v + 0x4B000000);" in src
        fn = "uchar root(int m0) {\n  const int m = m0 + 0x4B000000;\n" + body + "}"
        n = 1 << 21
        m = np.arange(n, dtype=np.int32)
        got = S.Map(c, fn, S.I32, S.U8)(S.Vector.from_numpy(c, m)).to_numpy()
        ref = np.minimum(np.sqrt(m.astype(np.float32)).astype(np.int64), 255).astype(np.uint8)
        assert np.array_equal(got, ref)
    finally:
        c.finalize()


def test_sobel_both_forms_full_image():
    """8192^2 (the bench's workload): the tuned user function and Listing 1.5
    give the oracle's whole image bit for bit"""
    c = tma_ctx()
    try:
        R = Cc = 8192
        img = I.image_u8(I.SEED_SOBEL, R, Cc)
        m = S.Matrix.from_numpy(c, img)
        ref = O.mapoverlap2d(O.OS_SOBEL, img, 1, O.OB_NEUTRAL, 0)
        for src in (A.SOBEL, A.SOBEL_TUNED):
            assert np.array_equal(S.MapOverlap(c, src, S.U8, S.U8, 1, S.NEUTRAL, 0)(m).to_numpy(), ref)
    finally:
        c.finalize()


@pytest.mark.parametrize("cw,rh,kt,full", [(16, 4, 2, -1), (8, 8, 1, -1), (4, 16, 1, -1), (8, 4, 1, -1),
                                           (16, 2, 2, -1), (8, 16, 1, 1), (8, 32, 1, 1), (8, 8, 2, 0),
                                           (16, 4, 1, 1)])
def test_sobel_tuned_geometries(cw, rh, kt, full):
    """the tuned Sobel in the register-block geometries the bench sweeps (with and
    without the unguarded full-tile loop, option mo_full), on a ragged 1000 x
    1500 image with every edge: bit-exact against the oracle"""
    c = tma_ctx()
    try:
        for k, v in (("mo_cw", cw), ("mo_rh", rh), ("mo_kt", kt), ("mo_full", full)):
            c.set_option(k, v)
        img = I.image_u8(I.SEED_SOBEL + 11, 1000, 1500)
        got = S.MapOverlap(c, A.SOBEL_TUNED, S.U8, S.U8, 1, S.NEUTRAL, 0)(S.Matrix.from_numpy(c, img)).to_numpy()
        assert np.array_equal(got, O.mapoverlap2d(O.OS_SOBEL, img, 1, O.OB_NEUTRAL, 0))
    finally:
        c.finalize()


@pytest.mark.parametrize("full", [0, 1])
@pytest.mark.parametrize("shape", [(37, 48), (65, 144), (513, 1008), (70, 1040)])
def test_full_tile_loop_forced(shape, full):
    """option mo_full forces the unguarded full-tile loop on (or off) whatever the
    tiles per block: byte and float stencils on ragged shapes stay bit-exact (the
    loop runs only for threads whose rows and packed stores are all in range)"""
    c = tma_ctx(mo_full=full, mo_kt=1)
    try:
        x8 = I.image_u8(I.SEED_SOBEL + 3, *shape)
        for src, kind in ((A.SOBEL, O.OS_SOBEL), (A.SOBEL_TUNED, O.OS_SOBEL), (A.IDENT2D_U8, O.OS_IDENT)):
            got = S.MapOverlap(c, src, S.U8, S.U8, 1, S.NEUTRAL, 0)(S.Matrix.from_numpy(c, x8)).to_numpy()
            assert np.array_equal(got, O.mapoverlap2d(kind, x8, 1, O.OB_NEUTRAL, 0)), (src, shape)
        x32 = I.image_f32(I.SEED_GAUSS + 3, shape[0], shape[1] // 4 * 4)
        got = S.MapOverlap(c, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)(S.Matrix.from_numpy(c, x32)).to_numpy()
        assert np.array_equal(got, O.mapoverlap2d(O.OS_GAUSS5, x32, 2, O.OB_NEAREST, 0.0))
    finally:
        c.finalize()


def test_sobel_tuned_bench_geometry_full_image():
    """8192^2 in the bench's sobel_tuned configuration (8 x 8 register block, one
    tile per block, the unguarded full-tile loop; also 16 x 8): the oracle's
    whole image"""
    for rh in (8, 16):
        _sobel_tuned_full_image(rh)


def _sobel_tuned_full_image(rh):
    c = tma_ctx(mo_rh=rh, mo_cw=8, mo_kt=1, mo_full=1)
    try:
        img = I.image_u8(I.SEED_SOBEL, 8192, 8192)
        got = S.MapOverlap(c, A.SOBEL_TUNED, S.U8, S.U8, 1, S.NEUTRAL, 0)(S.Matrix.from_numpy(c, img)).to_numpy()
        assert np.array_equal(got, O.mapoverlap2d(O.OS_SOBEL, img, 1, O.OB_NEUTRAL, 0))
    finally:
        c.finalize()
