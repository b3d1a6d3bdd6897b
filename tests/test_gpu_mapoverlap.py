"""GPU parity tests for MapOverlap: bit-exact against the oracle
(same operation order, -fmad=false), both boundary modes, matrix and vector
forms, tile-ragged sizes, and the get() bounds check (A21)."""
import numpy as np
import pytest

import oracle as O
from gpu_util import require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu

SHAPES = [(1, 1), (2, 3), (37, 53), (64, 128), (65, 129), (200, 300), (513, 1000)]


@pytest.fixture(scope="module")
def ctx():
    require_gpu()
    c = S.Context(1)
    yield c
    c.finalize()


@pytest.fixture(scope="module")
def mo(ctx):
    return dict(
        box_n=S.MapOverlap(ctx, A.BOX3, S.F32, S.F32, 1, S.NEUTRAL, 0.0),
        box_c=S.MapOverlap(ctx, A.BOX3, S.F32, S.F32, 1, S.NEAREST, 0.0),
        sobel=S.MapOverlap(ctx, A.SOBEL, S.U8, S.U8, 1, S.NEUTRAL, 0),
        gauss=S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0),
        gauss_n=S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEUTRAL, 0.0),
        sx=S.MapOverlap(ctx, A.SHIFTX, S.F32, S.F32, 1, S.NEUTRAL, 7.0),
        sy=S.MapOverlap(ctx, A.SHIFTY, S.F32, S.F32, 1, S.NEAREST, 0.0),
        sxu=S.MapOverlap(ctx, A.SHIFTX_U8, S.U8, S.U8, 1, S.NEAREST, 0),
        id1=S.MapOverlap(ctx, A.IDENT1D, S.F32, S.F32, 1, S.NEUTRAL, 0.0),
        sh1=S.MapOverlap(ctx, A.SHIFT1D, S.F32, S.F32, 1, S.NEUTRAL, -1.0),
        box1=S.MapOverlap(ctx, A.BOX1D, S.F32, S.F32, 1, S.NEAREST, 0.0),
    )


def mat(ctx, a):
    return S.Matrix.from_numpy(ctx, a)


@pytest.mark.parametrize("shape", SHAPES)
def test_box_sum_listing_1_2(ctx, mo, shape):
    x = I.image_f32(41, *shape)
    m = mat(ctx, x)
    assert np.array_equal(mo["box_n"](m).to_numpy(), O.mapoverlap2d(O.OS_BOX3, x, 1, O.OB_NEUTRAL, 0.0))
    assert np.array_equal(mo["box_c"](m).to_numpy(), O.mapoverlap2d(O.OS_BOX3, x, 1, O.OB_NEAREST, 0.0))


def test_golden_boxsum_and_sobel(ctx, mo, golden):
    g = golden("boxsum_4x4.txt")
    x = np.array(g["input"], np.float32)
    assert np.array_equal(mo["box_n"](mat(ctx, x)).to_numpy(), np.array(g["output"], np.float32))
    g = golden("sobel_impulse_5x5.txt")
    x = np.array(g["input"], np.uint8)
    assert np.array_equal(mo["sobel"](mat(ctx, x)).to_numpy(), np.array(g["output"], np.uint8))


@pytest.mark.parametrize("shape", SHAPES + [(8, 8192)])
def test_sobel_bitexact(ctx, mo, shape):
    x = I.image_u8(I.SEED_SOBEL, *shape)
    assert np.array_equal(mo["sobel"](mat(ctx, x)).to_numpy(), O.mapoverlap2d(O.OS_SOBEL, x, 1, O.OB_NEUTRAL, 0))


@pytest.mark.parametrize("shape", SHAPES)
def test_gaussian_bitexact(ctx, mo, shape):
    x = I.image_f32(I.SEED_GAUSS, *shape)
    m = mat(ctx, x)
    assert np.array_equal(mo["gauss"](m).to_numpy(), O.mapoverlap2d(O.OS_GAUSS5, x, 2, O.OB_NEAREST, 0.0))
    assert np.array_equal(mo["gauss_n"](m).to_numpy(), O.mapoverlap2d(O.OS_GAUSS5, x, 2, O.OB_NEUTRAL, 0.0))


def test_orientation_dx_is_column(ctx, mo):
    x = I.image_f32(42, 37, 53)
    assert np.array_equal(mo["sx"](mat(ctx, x)).to_numpy(), O.mapoverlap2d(O.OS_SHIFT_X, x, 1, O.OB_NEUTRAL, 7.0))
    assert np.array_equal(mo["sy"](mat(ctx, x)).to_numpy(), O.mapoverlap2d(O.OS_SHIFT_Y, x, 1, O.OB_NEAREST, 0.0))
    xu = I.image_u8(43, 9, 11)
    assert np.array_equal(mo["sxu"](mat(ctx, xu)).to_numpy(), O.mapoverlap2d(O.OS_SHIFT_X, xu, 1, O.OB_NEAREST, 0))


@pytest.mark.parametrize("n", [1, 2, 100, 1023, 1024, 1025, 100001])
def test_mapoverlap_vector(ctx, mo, n):
    v = I.uniform_f32(44, n)
    vv = S.Vector.from_numpy(ctx, v)
    assert np.array_equal(mo["id1"](vv).to_numpy(), O.mapoverlap1d(O.OS_IDENT, v, 1, O.OB_NEUTRAL, 0.0))
    assert np.array_equal(mo["sh1"](vv).to_numpy(), O.mapoverlap1d(O.OS_SHIFT_X, v, 1, O.OB_NEUTRAL, -1.0))
    assert np.array_equal(mo["box1"](vv).to_numpy(), O.mapoverlap1d(O.OS_BOX3, v, 1, O.OB_NEAREST, 0.0))


def test_iterated_stencil(ctx, mo):
    # output (block, with halo room) feeds the next MapOverlap: halo refresh path
    x = I.image_f32(45, 130, 70)
    a = mat(ctx, x)
    b = mo["gauss"](a)
    c = mo["gauss"](b)
    r1 = O.mapoverlap2d(O.OS_GAUSS5, x, 2, O.OB_NEAREST, 0.0)
    assert np.array_equal(c.to_numpy(), O.mapoverlap2d(O.OS_GAUSS5, r1, 2, O.OB_NEAREST, 0.0))


def test_debug_bounds_flags_access_beyond_d():
    require_gpu()
    with S.Context(1) as c:
        c.set_option("debug_bounds", 1)
        # an offset the static check cannot prove (a runtime value) -> runtime check
        bad = S.MapOverlap(c, "float f(const float* p){ int k = (int)(p[0] * 0.0f) + 2; return get(p, k, 0); }",
                           S.F32, S.F32, 1)
        assert not bad.bounds_proven
        with pytest.raises(S.SklError) as e:
            bad(S.Matrix.from_numpy(c, np.ones((8, 8), np.float32)))
        assert e.value.name == "OUT_OF_RANGE"
        ok = S.MapOverlap(c, A.BOX3, S.F32, S.F32, 1, S.NEUTRAL, 0.0)
        x = np.ones((8, 8), np.float32)
        assert np.array_equal(ok(S.Matrix.from_numpy(c, x)).to_numpy(),
                              O.mapoverlap2d(O.OS_BOX3, x, 1, O.OB_NEUTRAL, 0.0))


@pytest.mark.parametrize("shape", [(5, 9), (131, 257), (600, 1030)])
def test_persistent_variant_bitexact(shape):
    """mo_persist=1 (resident blocks walking the tiles with two staging buffers;
    measured slower on B200, kept selectable) gives the oracle's results"""
    require_gpu()
    c = S.Context(1)
    try:
        c.set_option("mo_persist", 1)
        img8 = I.image_u8(I.SEED_SOBEL, *shape)
        sob = S.MapOverlap(c, A.SOBEL, S.U8, S.U8, 1, S.NEUTRAL, 0)
        assert np.array_equal(sob(S.Matrix.from_numpy(c, img8)).to_numpy(),
                              O.mapoverlap2d(O.OS_SOBEL, img8, 1, O.OB_NEUTRAL, 0))
        imgf = I.image_f32(I.SEED_GAUSS, *shape)
        gau = S.MapOverlap(c, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
        assert np.array_equal(gau(S.Matrix.from_numpy(c, imgf)).to_numpy(),
                              O.mapoverlap2d(O.OS_GAUSS5, imgf, 2, O.OB_NEAREST, 0.0))
    finally:
        c.finalize()
