"""Every Scan schedule the library ships (skl_set_option "scan_variant"), not
only the default, against the oracle: int32 bit-exact, fp32
within 1e-5, and the non-commutative affine composition (operand order, A10)
bit-exact; sizes span many tiles plus ragged tails, tile sizes 2-16 chunks."""
import numpy as np
import pytest

import oracle as O
from gpu_util import rel_l2, require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu

# (variant, block_threads, scan_chunks): 6 = default (tile in shared memory),
# 3 = items in registers, 2 = warp-wide look-back, 4 = persistent pipeline,
# 0 = persistent chunked
CONFIGS = [(6, 256, 8), (6, 128, 16), (6, 256, 2), (3, 256, 8), (2, 128, 4), (4, 256, 8), (0, 256, 8)]
SIZES = [1, 7, 2048, 8193, 65536 * 3 + 11, (1 << 22) + 5]


@pytest.fixture(scope="module", params=CONFIGS, ids=lambda c: f"v{c[0]}b{c[1]}c{c[2]}")
def sk(request):
    require_gpu()
    var, bt, ch = request.param
    c = S.Context(1)
    c.set_option("scan_variant", var)
    c.set_option("block_threads", bt)
    c.set_option("scan_chunks", ch)
    aff = c.struct_type("Aff", A.AFFINE_DECL, 8, 4)
    d = dict(ctx=c, aff=aff, f=S.Scan(c, A.ADD, S.F32), i=S.Scan(c, A.ADD_I32, S.I32),
             a=S.Scan(c, A.AFFINE_COMPOSE, aff), l=S.Scan(c, A.LEFT_F32, S.F32))
    yield d
    c.finalize()


@pytest.mark.parametrize("n", SIZES)
def test_scan_variant(sk, n):
    ctx = sk["ctx"]
    xi = I.uniform_int(71, n, -1000, 1000)
    assert np.array_equal(sk["i"](S.Vector.from_numpy(ctx, xi)).to_numpy(), O.scan(O.OP_ADD_I32, xi))
    x = I.uniform_f32(72, n)
    v = S.Vector.from_numpy(ctx, x)
    assert rel_l2(sk["f"](v).to_numpy(), O.scan(O.OP_ADD_F32, x)) <= 1e-5
    assert np.array_equal(sk["l"](v).to_numpy(), O.scan(O.OP_LEFT_F32, x))
    if n <= 300000:
        p = I.uniform_int(73, 2 * n, 0, 2**32 - 1, np.uint64).astype(np.uint32).reshape(n, 2)
        got = sk["a"](S.Vector(ctx, sk["aff"], n).copy_in(p)).to_numpy(np.uint32).reshape(n, 2)
        assert np.array_equal(got, O.scan(O.OP_AFFINE_U32, p))


def test_repeated_calls_reuse_status(sk):
    """the status words are reused across calls via epochs (no reset kernel)"""
    ctx = sk["ctx"]
    xi = I.uniform_int(74, 100003, -5, 5)
    v = S.Vector.from_numpy(ctx, xi)
    want = O.scan(O.OP_ADD_I32, xi)
    out = sk["i"](v)
    for _ in range(5):
        sk["i"](v, out=out)
        assert np.array_equal(out.to_numpy(), want)
