"""The one-process-per-GPU mode (skl_init_dist: NCCL communicator, collective
host reads, rank-local parts) exercised on one GPU with world size 1, so that
its code paths run on real hardware even where only one GPU is available; the
exchange logic itself is covered by tests/test_dist_gloo.py (2 ranks)."""
import numpy as np
import pytest

import oracle as O
from gpu_util import rel_l2, require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def ctx():
    require_gpu()
    c = S.Context.dist(0, 1, 0, S.Context.nccl_unique_id())
    yield c
    c.finalize()


def test_dist_context_shape(ctx):
    assert ctx.devices() == (1, 0, 1)


def test_skeletons_in_dist_mode(ctx):
    n = 100003
    a, b = I.uniform_f32(I.SEED_DOT_A, n), I.uniform_f32(I.SEED_DOT_B, n)
    va, vb = S.Vector.from_numpy(ctx, a), S.Vector.from_numpy(ctx, b)
    got = float(S.Reduce(ctx, A.SUM, S.F32)(S.Zip(ctx, A.MULT, S.F32, S.F32, S.F32)(va, vb)).scalar())
    ref = O.reduce_(O.OP_ADD_F32, O.zip_(O.OZ_MULT_F32, a, b))
    assert abs(got - ref) <= 1e-5 * abs(ref)
    xi = I.uniform_int(3, n, -1000, 1000)
    assert np.array_equal(S.Scan(ctx, A.ADD_I32, S.I32)(S.Vector.from_numpy(ctx, xi)).to_numpy(),
                          O.scan(O.OP_ADD_I32, xi))
    img = I.image_u8(I.SEED_SOBEL, 67, 129)
    sob = S.MapOverlap(ctx, A.SOBEL, S.U8, S.U8, 1, S.NEUTRAL, 0)
    s1 = sob(S.Matrix.from_numpy(ctx, img))
    r1 = O.mapoverlap2d(O.OS_SOBEL, img, 1, O.OB_NEUTRAL, 0)
    assert np.array_equal(sob(s1).to_numpy(), O.mapoverlap2d(O.OS_SOBEL, r1, 1, O.OB_NEUTRAL, 0))


def test_distributions_in_dist_mode(ctx):
    x = I.uniform_f32(9, 4097)
    v = S.Vector.from_numpy(ctx, x)
    for d in (S.BLOCK, S.COPY, S.BLOCK):
        v.set_distribution(d)
        assert np.array_equal(v.to_numpy(), x)
    v.set_distribution(S.SINGLE, 0)
    assert np.array_equal(v.to_numpy(), x)
    addf = S.Reduce(ctx, A.ADD, S.F32)
    c = S.Vector(ctx, S.F32, 1000).set_distribution(S.COPY, 0, addf)
    c.fill(2.0)
    c.set_distribution(S.BLOCK)          # copy(+) -> block with one replica
    assert np.array_equal(c.to_numpy(), np.full(1000, 2.0, np.float32))


def test_lmosem_subset_in_dist_mode(ctx):
    from paper_conf_pact_steuwerg13_b200.lmosem import ListModeOSEM
    N, nev = 12, 4000
    events = I.lmosem_events(I.SEED_LMOSEM, nev, N)
    f0 = np.ones(N ** 3, np.float32)
    osem = ListModeOSEM(ctx, N)
    osem.load_events(events, 2)
    osem.set_image(f0)
    osem.iterate(1)
    f = f0
    for lo, hi in ListModeOSEM.subset_bounds(nev, 2):
        f = O.lmosem(events[lo:hi], N, f)[1].astype(np.float32)
    assert rel_l2(osem.image(), f) <= 1e-4
    osem.destroy()
