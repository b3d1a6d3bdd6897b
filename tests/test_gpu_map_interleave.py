"""The warp-interleaved Map/Zip kernel (skl_set_option "map_interleave" 1:
lane l of a warp handles elements base + j*32 + l) against the oracle, bit-exact,
for every element width, ragged sizes, Zip, a void Map with extra arguments
(LM OSEM) and Mandelbrot."""
import numpy as np
import pytest

import oracle as O
from gpu_util import rel_l2, require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu

SIZES = [1, 31, 33, 1000, 4097, (1 << 20) + 3]


@pytest.fixture(scope="module", params=[(256, 1, 0), (1024, 1, 0), (128, 4, 0), (128, 1, 1), (64, 1, 3)],
                ids=lambda p: f"b{p[0]}u{p[1]}j{p[2]}")
def ctx(request):
    require_gpu()
    bt, un, j = request.param
    c = S.Context(1)
    c.set_option("map_interleave", 1)
    c.set_option("block_threads", bt)
    c.set_option("map_unroll", un)
    c.set_option("map_il_elems", j)   # elements per lane (0 = one chunk)
    yield c
    c.finalize()


@pytest.mark.parametrize("n", SIZES)
def test_map_zip_interleaved(ctx, n):
    x = I.uniform_f32(41, n) - np.float32(0.5)
    assert np.array_equal(S.Map(ctx, A.SQP1, S.F32, S.F32)(S.Vector.from_numpy(ctx, x)).to_numpy(),
                          O.map_(O.OM_SQP1_F32, x))
    u = I.uniform_int(42, n, 0, 255, np.int64).astype(np.uint8)
    assert np.array_equal(S.Map(ctx, A.INV_U8, S.U8, S.U8)(S.Vector.from_numpy(ctx, u)).to_numpy(),
                          O.map_(O.OM_INV_U8, u))
    y = I.uniform_f32(43, n)
    z = S.Zip(ctx, A.ADD, S.F32, S.F32, S.F32)(S.Vector.from_numpy(ctx, x), S.Vector.from_numpy(ctx, y))
    assert np.array_equal(z.to_numpy(), O.zip_(O.OZ_ADD_F32, x, y))


@pytest.mark.parametrize("block", [1, 7, 12, 16])
def test_mandelbrot_blocktest_exact(ctx, block, golden):
    """the amortised escape test (apps.mandelbrot_blocktest) gives the oracle's
    counts: a coarse grid of the A22 window, the hand-derived golden points
    (including c = -2, whose orbit stays at |z| = 2 exactly), points just outside
    |c| = 2 in the window's corners, and MAX values that are not multiples of the
    block"""
    gp = np.array(golden("mandelbrot_points.txt")[None], np.float64)   # re, im, count (MAX 1000)
    pts = gp[:, :2].astype(np.float32)
    grid = I.mandel_grid(48, 64)
    extra = np.array([[-2.0, 1.125], [-2.0, -1.125], [0.99, 1.12], [-0.75, 0.1], [0.2501, 0.0]], np.float32)
    cs = np.concatenate([pts, extra, grid.reshape(-1, 2)])
    for mx in (1000, 37):
        m = S.Map(ctx, A.mandelbrot_blocktest(mx, block), S.F32X2, S.U32)
        got = m(S.Matrix(ctx, S.F32X2, 1, cs.shape[0]).copy_in(cs[None])).to_numpy().ravel()
        assert np.array_equal(got, O.mandelbrot(cs[None], mx)[0].ravel()), (block, mx)
        if mx == 1000:
            assert np.array_equal(got[:len(gp)], gp[:, 2].astype(np.uint32))


def test_mandelbrot_interleaved(ctx):
    R, C = 96, 128
    grid = I.mandel_grid(R, C)      # a coarse 96 x 128 view of the A22 window
    m = S.Map(ctx, A.mandelbrot_blocktest(1000, 12), S.F32X2, S.U32)
    got = m(S.Matrix(ctx, S.F32X2, R, C).copy_in(grid)).to_numpy()
    ref, _ = O.mandelbrot(grid, 1000)
    assert np.array_equal(got, ref)


def test_void_map_with_extras_interleaved(ctx):
    N, nev = 12, 5000
    evd = ctx.struct_type("Event", A.EVENT_DECL, A.EVENT_SIZE, 4)
    lm = S.Map(ctx, A.lmosem_map(N), evd, S.VOID, extra=[S.F32 | S.PTR, S.F32 | S.PTR])
    addf = S.Reduce(ctx, A.ADD, S.F32)
    events = I.lmosem_events(I.SEED_LMOSEM, nev, N)
    f0 = np.ones(N ** 3, np.float32)
    ev = S.Vector(ctx, evd, nev).copy_in(events).set_distribution(S.BLOCK)
    f = S.Vector.from_numpy(ctx, f0).set_distribution(S.COPY)
    c = S.Vector(ctx, S.F32, N ** 3).set_distribution(S.COPY, 0, addf)
    c.fill(0.0)
    lm(ev, f, (c, S.WRITE))
    c_ref, _, _, _ = O.lmosem(events, N, f0)
    assert rel_l2(c.to_numpy(), c_ref) <= 1e-4
