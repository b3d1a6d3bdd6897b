"""Allpairs on the GPU vs the oracle: both forms (row function;
zip + reduce), bit-exact (every C element is folded over k in order in fp32,
-fmad=false, as the oracle does), ragged tile edges, block(A) x copy(B) on
several logical devices."""
import numpy as np
import pytest

import oracle as O
from gpu_util import require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu

# d % 4 == 0 (4-byte inputs) takes the 128 x 128 kernel (d = 4: tail slice only;
# d = 20, 36, 100: full slices + tail); other d the 64 x 64 one
SHAPES = [(1, 1, 1), (2, 3, 3), (70, 33, 13), (130, 200, 64), (257, 129, 100), (64, 64, 16), (5, 300, 4),
          (129, 257, 20), (300, 130, 36), (256, 384, 32)]


@pytest.fixture(scope="module", params=[1, 3])
def ctx(request):
    require_gpu()
    G = request.param
    c = S.Context(G, devices=[0] * G)
    yield c
    c.finalize()


@pytest.fixture(scope="module")
def sk(ctx):
    return dict(
        man=S.Allpairs(ctx, A.MANHATTAN_ROWS, S.F32, S.F32),
        dot=S.Allpairs(ctx, A.DOT_ROWS, S.F32, S.F32),
        man_zr=S.Allpairs(ctx, A.ABSDIFF, S.F32, S.F32, reduce=A.ADD),
        dot_zr=S.Allpairs(ctx, A.MULT, S.F32, S.F32, reduce=A.ADD),
    )


@pytest.mark.parametrize("shape", SHAPES)
def test_allpairs_bitexact(ctx, sk, shape):
    n, m, d = shape
    a = I.uniform_f32(81, n * d).reshape(n, d) - np.float32(0.5)
    b = I.uniform_f32(82, m * d).reshape(m, d) - np.float32(0.5)
    ma = S.Matrix.from_numpy(ctx, a).set_distribution(S.BLOCK)
    mb = S.Matrix.from_numpy(ctx, b)
    man = O.allpairs(O.AP_MANHATTAN, a, b)
    dot = O.allpairs(O.AP_DOT, a, b)
    assert np.array_equal(sk["man"](ma, mb).to_numpy(), man)
    assert np.array_equal(sk["dot"](ma, mb).to_numpy(), dot)
    assert np.array_equal(sk["man_zr"](ma, mb).to_numpy(), man)
    c = sk["dot_zr"](ma, mb)
    assert c.distribution()[0] == S.BLOCK
    assert np.array_equal(c.to_numpy(), dot)


def test_golden_and_eq2(ctx, sk, golden):
    g = golden("allpairs_small.txt")
    a, b = np.array(g["A"], np.float32), np.array(g["B"], np.float32)
    ma, mb = S.Matrix.from_numpy(ctx, a), S.Matrix.from_numpy(ctx, b)
    assert np.array_equal(sk["dot_zr"](ma, mb).to_numpy(), np.array(g["dot"], np.float32))
    assert np.array_equal(sk["man"](ma, mb).to_numpy(), np.array(g["manhattan"], np.float32))
    # Eq. (2): A x B = allpairs(dotProduct)(A, B^T)
    x = I.uniform_f32(83, 96 * 40).reshape(96, 40)
    y = I.uniform_f32(84, 40 * 72).reshape(40, 72)
    c = sk["dot_zr"](S.Matrix.from_numpy(ctx, x), S.Matrix.from_numpy(ctx, np.ascontiguousarray(y.T))).to_numpy()
    assert np.allclose(c, x.astype(np.float64) @ y.astype(np.float64), rtol=1e-5, atol=1e-5)


def test_size_mismatch(ctx, sk):
    with pytest.raises(S.SklError) as e:
        sk["man"](S.Matrix.from_numpy(ctx, np.zeros((3, 4), np.float32)),
                  S.Matrix.from_numpy(ctx, np.zeros((3, 5), np.float32)))
    assert e.value.name == "SIZE_MISMATCH"


@pytest.mark.parametrize("tile", [2, 4, 8])
def test_forced_tile_widths_bitexact(ctx, sk, tile):
    """the 128-row kernels (128 x 64 and 128 x 128 tiles of C, and the hybrid of
    both, here with every tile split) agree with the oracle"""
    ctx.set_option("ap_tile", tile)
    try:
        for n, m, d in ((130, 200, 64), (257, 129, 100), (5, 300, 4)):
            a = I.uniform_f32(85, n * d).reshape(n, d)
            b = I.uniform_f32(86, m * d).reshape(m, d)
            ma, mb = S.Matrix.from_numpy(ctx, a), S.Matrix.from_numpy(ctx, b)
            assert np.array_equal(sk["dot_zr"](ma, mb).to_numpy(), O.allpairs(O.AP_DOT, a, b))
            assert np.array_equal(sk["man_zr"](ma, mb).to_numpy(), O.allpairs(O.AP_MANHATTAN, a, b))
    finally:
        ctx.set_option("ap_tile", 0)


def test_hybrid_last_wave_bitexact(ctx, sk):
    """automatic hybrid: 18 x 18 = 324 tiles of 128 x 128 on one device leave the
    last wave (296 slots) 28 tiles deep, which run as 56 halves of 128 x 64;
    ragged n and m put some halves partly or wholly beyond the matrix"""
    G = ctx.ndev
    for n, m, d in ((2304 * G, 2304, 8), (2300 * G - 3, 2290, 12)):
        a = I.uniform_f32(87, n * d).reshape(n, d) - np.float32(0.5)
        b = I.uniform_f32(88, m * d).reshape(m, d) - np.float32(0.5)
        ma = S.Matrix.from_numpy(ctx, a).set_distribution(S.BLOCK)
        mb = S.Matrix.from_numpy(ctx, b)
        assert np.array_equal(sk["dot_zr"](ma, mb).to_numpy(), O.allpairs(O.AP_DOT, a, b))
        assert np.array_equal(sk["man_zr"](ma, mb).to_numpy(), O.allpairs(O.AP_MANHATTAN, a, b))


@pytest.mark.parametrize("tile", [0, 4, 8])
def test_k_slice_32_bitexact(ctx, sk, tile):
    """32-deep k-slices (ap_bk=32, dynamic shared memory): d below one slice,
    one slice plus a tail, several slices plus a tail"""
    ctx.set_option("ap_bk", 32)
    ctx.set_option("ap_tile", tile)
    try:
        sk2 = S.Allpairs(ctx, A.MULT, S.F32, S.F32, reduce=A.ADD)
        for n, m, d in ((130, 200, 20), (257, 129, 36), (129, 300, 100), (64, 64, 64)):
            a = I.uniform_f32(89, n * d).reshape(n, d) - np.float32(0.5)
            b = I.uniform_f32(90, m * d).reshape(m, d) - np.float32(0.5)
            ma, mb = S.Matrix.from_numpy(ctx, a), S.Matrix.from_numpy(ctx, b)
            assert np.array_equal(sk2(ma, mb).to_numpy(), O.allpairs(O.AP_DOT, a, b))
    finally:
        ctx.set_option("ap_bk", 0)
        ctx.set_option("ap_tile", 0)
