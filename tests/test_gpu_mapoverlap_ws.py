"""GPU parity tests for the TMA / warp-specialised 2-D MapOverlap kernel
(mo_ws=1): a producer warp stages each tile with one
cp.async.bulk.tensor copy (out-of-matrix cells zero-filled, then patched for
NEAREST and non-zero NEUTRAL, A20) and the consumer warps apply f.
Bit-exact against the oracle at sizes spanning several tiles with ragged
edges, every boundary mode, several ring depths, logical multi-device runs
(overlap distribution: the TMA map covers a part with halo rows) and the fused
halo push."""
import numpy as np
import pytest

import oracle as O
from gpu_util import require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu

SHAPES = [(1, 4), (3, 16), (37, 52), (65, 132), (200, 300), (513, 1000)]
SHAPES_U8 = [(1, 16), (3, 32), (37, 48), (65, 144), (200, 304), (513, 1008)]   # rows of 16-byte multiples


def ws_ctx(ndev=1, **opts):
    require_gpu()
    c = S.Context(ndev, devices=[0] * ndev)
    c.set_option("mo_ws", 1)
    for k, v in opts.items():
        c.set_option(k, v)
    return c


@pytest.mark.parametrize("shape", SHAPES)
@pytest.mark.parametrize("stages", [2, 4])
def test_ws_f32_modes(shape, stages):
    c = ws_ctx(mo_ws_stages=stages)
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
        assert c.counter("tma_launches") - before == 5   # every call took the TMA kernel
    finally:
        c.finalize()


@pytest.mark.parametrize("shape", SHAPES_U8)
def test_ws_u8_sobel_and_shift(shape):
    # u8 tiles need a staged row <= 256 bytes: 4 outputs per thread and row
    c = ws_ctx(mo_cw=4)
    try:
        x = I.image_u8(I.SEED_SOBEL, *shape)
        m = S.Matrix.from_numpy(c, x)
        before = c.counter("tma_launches")
        sob = S.MapOverlap(c, A.SOBEL, S.U8, S.U8, 1, S.NEUTRAL, 0)
        assert np.array_equal(sob(m).to_numpy(), O.mapoverlap2d(O.OS_SOBEL, x, 1, O.OB_NEUTRAL, 0))
        sx = S.MapOverlap(c, A.SHIFTX_U8, S.U8, S.U8, 1, S.NEAREST, 0)
        assert np.array_equal(sx(m).to_numpy(), O.mapoverlap2d(O.OS_SHIFT_X, x, 1, O.OB_NEAREST, 0))
        assert c.counter("tma_launches") - before == 2
    finally:
        c.finalize()


def test_ws_u8_wide_rows():
    """16 outputs per thread make the staged u8 row 544 bytes: described in 8-byte
    units (68 <= 256) the tile still goes through TMA"""
    c = ws_ctx()
    try:
        x = I.image_u8(I.SEED_SOBEL, 70, 608)
        sob = S.MapOverlap(c, A.SOBEL, S.U8, S.U8, 1, S.NEUTRAL, 0)
        before = c.counter("tma_launches")
        assert np.array_equal(sob(S.Matrix.from_numpy(c, x)).to_numpy(),
                              O.mapoverlap2d(O.OS_SOBEL, x, 1, O.OB_NEUTRAL, 0))
        assert c.counter("tma_launches") == before + 1
    finally:
        c.finalize()


def test_ws_unaligned_rows_fall_back():
    """rows of 4 * 13 bytes are not 16-byte multiples (no TMA map): plain kernel"""
    c = ws_ctx()
    try:
        x = I.image_f32(I.SEED_GAUSS, 50, 13)
        gau = S.MapOverlap(c, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
        before = c.counter("tma_launches")
        assert np.array_equal(gau(S.Matrix.from_numpy(c, x)).to_numpy(),
                              O.mapoverlap2d(O.OS_GAUSS5, x, 2, O.OB_NEAREST, 0.0))
        assert c.counter("tma_launches") == before
    finally:
        c.finalize()


@pytest.mark.parametrize("ndev", [2, 3])
def test_ws_overlap_distribution_and_halo_push(ndev):
    """parts with halo rows (the TMA map starts at the part's first row), and an
    iterated stencil whose halos are pushed by the kernel"""
    c = ws_ctx(ndev)
    try:
        x = I.image_f32(I.SEED_GAUSS, 301, 260)
        gau = S.MapOverlap(c, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
        a = S.Matrix.from_numpy(c, x)
        b = gau(a)
        t = gau(b)
        ref = x
        for _ in range(2):
            ref = O.mapoverlap2d(O.OS_GAUSS5, ref, 2, O.OB_NEAREST, 0.0)
        assert np.array_equal(t.to_numpy(), ref)
        assert c.counter("tma_launches") >= 2 * ndev
    finally:
        c.finalize()
