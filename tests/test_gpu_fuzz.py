"""Randomised coherence test: seeded random programs of container operations on
1-3 logical devices, checked against a numpy shadow of every container after
every read.  It exercises the interplay of the state the library keeps per
container: distributions and redistribution, lazy (deferred) Map/Zip results and
their fusion into Reduce, chunked uploads consumed by Maps, pushed halos of
MapOverlap outputs, host mirrors, in-place calls, unaligned views (parts that
keep halo room after overlap -> block), Scan and 1-D stencils.  Bit-exact except
the fp32 Reduce and Scan (relative 1e-5)."""
import numpy as np
import pytest

import oracle as O
from gpu_util import require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu

SIZES = [(1 << 20) + 7, 4099, 3]          # the first one is chunked on upload (>= 4 MB)
ROWS, COLS = 130, 67                        # matrix shape for the stencils


def _no_overlap(c):
    """an in-place Map/Zip needs a block/copy/single input (the output of an
    elementwise skeleton has no halo)"""
    if c.distribution()[0] == S.OVERLAP:
        c.set_distribution(S.BLOCK)


def _program(G, seed, steps=60):
    rng = np.random.default_rng(seed)
    ctx = S.Context(G, devices=[0] * G)
    try:
        neg = S.Map(ctx, A.NEG, S.F32, S.F32)
        sq = S.Map(ctx, A.SQP1, S.F32, S.F32)
        add = S.Zip(ctx, A.ADD, S.F32, S.F32, S.F32)
        red = S.Reduce(ctx, A.SUM, S.F32)
        box = S.MapOverlap(ctx, A.BOX3, S.F32, S.F32, 1, S.NEAREST, 0.0)
        box1 = S.MapOverlap(ctx, A.BOX1D, S.F32, S.F32, 1, S.NEAREST, 0.0)
        scan = S.Scan(ctx, A.ADD, S.F32)
        n = SIZES[rng.integers(len(SIZES))]
        vecs = [S.Vector(ctx, S.F32, n) for _ in range(3)]
        shadow = [np.zeros(n, np.float32) for _ in range(3)]
        for v in vecs:
            v.fill(0.0)
        mat = [S.Matrix(ctx, S.F32, ROWS, COLS) for _ in range(2)]
        mshadow = [np.zeros((ROWS, COLS), np.float32) for _ in range(2)]
        for m in mat:
            m.fill(0.0)
        dists = [(S.BLOCK, 0), (S.COPY, 0), (S.SINGLE, G - 1), (S.OVERLAP, 1), (S.BLOCK, 0)]
        log = []
        for step in range(steps):
            op = int(rng.integers(14))
            i, j, k = (int(x) for x in rng.integers(3, size=3))
            log.append((op, i, j, k))
            if op == 0:        # host write
                x = (rng.random(n, dtype=np.float32) - np.float32(0.5))
                vecs[i].copy_in(x)
                shadow[i] = x
            elif op == 1:      # redistribution
                d, a = dists[int(rng.integers(len(dists)))]
                vecs[i].set_distribution(d, a)
            elif op == 2:      # Map into another container (or in place)
                f, ref = (neg, O.OM_NEG_F32) if rng.random() < 0.5 else (sq, O.OM_SQP1_F32)
                if i == j:
                    _no_overlap(vecs[i])
                f(vecs[i], out=vecs[j])
                shadow[j] = O.map_(ref, shadow[i])
            elif op == 3:      # Zip
                if k == i:
                    _no_overlap(vecs[i])
                add(vecs[i], vecs[j], out=vecs[k])
                shadow[k] = O.zip_(O.OZ_ADD_F32, shadow[i], shadow[j])
            elif op == 4:      # deferred chain read back on the host
                got = neg(sq(vecs[i])).to_numpy()
                assert np.array_equal(got, O.map_(O.OM_NEG_F32, O.map_(O.OM_SQP1_F32, shadow[i]))), log
            elif op == 5:      # Reduce of a deferred Zip (fused)
                got = float(red(add(vecs[i], vecs[j])).scalar())
                ref = O.reduce_(O.OP_ADD_F32, O.zip_(O.OZ_ADD_F32, shadow[i], shadow[j]))
                assert abs(got - ref) <= 1e-5 * max(1.0, float(np.abs(shadow[i]).sum() + np.abs(shadow[j]).sum())), log
            elif op == 6:      # read back
                assert np.array_equal(vecs[i].to_numpy(), shadow[i]), log
            elif op == 7:      # fill
                val = float(rng.integers(-3, 4))
                vecs[i].fill(val)
                shadow[i] = np.full(n, val, np.float32)
            elif op == 8:      # stencil ping-pong (pushed halos on G > 1)
                a, b = i % 2, 1 - i % 2
                box(mat[a], out=mat[b])
                mshadow[b] = O.mapoverlap2d(O.OS_BOX3, mshadow[a], 1, O.OB_NEAREST, 0.0)
            elif op == 9:      # matrix host write or Map on a matrix
                if rng.random() < 0.5:
                    x = rng.random((ROWS, COLS), dtype=np.float32)
                    mat[i % 2].copy_in(x)
                    mshadow[i % 2] = x
                else:
                    _no_overlap(mat[i % 2])
                    neg(mat[i % 2], out=mat[i % 2])
                    mshadow[i % 2] = -mshadow[i % 2]
            elif op == 10:     # matrix read back / redistribution
                if rng.random() < 0.5:
                    assert np.array_equal(mat[i % 2].to_numpy(), mshadow[i % 2]), log
                else:
                    d, a2 = dists[int(rng.integers(len(dists)))]
                    mat[i % 2].set_distribution(d, a2)
            elif op == 11:     # Scan (fp32: relative L2 against the double oracle)
                got = scan(vecs[i]).to_numpy().astype(np.float64)
                ref = O.scan(O.OP_ADD_F32, shadow[i])
                den = max(1e-30, float(np.linalg.norm(np.cumsum(np.abs(shadow[i].astype(np.float64))))))
                assert float(np.linalg.norm(got - ref)) <= 1e-5 * den, log
            elif op == 12:     # 1-D stencil into another vector
                if i != j:
                    box1(vecs[i], out=vecs[j])
                    shadow[j] = O.mapoverlap1d(O.OS_BOX3, shadow[i], 1, O.OB_NEAREST, 0.0)
            elif op == 13:     # a deferred chain materialised into an explicit output
                if i == j:
                    _no_overlap(vecs[i])
                neg(sq(vecs[i]), out=vecs[j])
                shadow[j] = O.map_(O.OM_NEG_F32, O.map_(O.OM_SQP1_F32, shadow[i]))
        for v, sh in zip(vecs, shadow):
            assert np.array_equal(v.to_numpy(), sh), log
        for m, sh in zip(mat, mshadow):
            assert np.array_equal(m.to_numpy(), sh), log
    finally:
        ctx.finalize()


@pytest.mark.parametrize("G", [1, 2, 3])
@pytest.mark.parametrize("seed", range(8))
def test_random_programs(G, seed):
    require_gpu()
    _program(G, 1000 * G + seed)
