"""Error behaviour of the C ABI on a GPU (include/skl.h conventions): every
failure is a negative status with a message, nothing aborts, and the context
stays usable afterwards."""
import numpy as np
import pytest

import oracle as O
from gpu_util import require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def ctx():
    require_gpu()
    c = S.Context(1)
    yield c
    c.finalize()


def _still_works(ctx):
    x = I.uniform_f32(11, 1001)
    neg = S.Map(ctx, A.NEG, S.F32, S.F32)
    assert np.array_equal(neg(S.Vector.from_numpy(ctx, x)).to_numpy(), O.map_(O.OM_NEG_F32, x))


def test_out_of_memory_is_reported(ctx):
    # 4 TiB, far beyond 180 GB of HBM; block-distributed so that fill() allocates
    # on the device (a host fill would try to pin 4 TiB of host memory)
    v = S.Vector(ctx, S.F32, 1 << 40).set_distribution(S.BLOCK)
    with pytest.raises(S.SklError) as e:
        v.fill(0.0)
    assert e.value.name == "OOM"
    v.destroy()
    _still_works(ctx)
    # the failed allocation must not resurface in a later launch check
    w = S.Vector(ctx, S.F32, 1 << 20).set_distribution(S.BLOCK)
    w.fill(1.0)
    assert float(S.Reduce(ctx, A.SUM, S.F32)(w).scalar()) == float(1 << 20)


def test_compile_error_carries_the_nvrtc_log(ctx):
    with pytest.raises(S.SklError) as e:
        S.Map(ctx, "float func(float x){ return x +* 2; }", S.F32, S.F32)
    assert e.value.name == "COMPILE"
    assert "error" in str(e.value).lower()
    _still_works(ctx)


def test_empty_and_mismatch(ctx):
    red = S.Reduce(ctx, A.SUM, S.F32)
    with pytest.raises(S.SklError) as e:
        red(S.Vector(ctx, S.F32, 0))
    assert e.value.name == "EMPTY"
    add = S.Zip(ctx, A.ADD, S.F32, S.F32, S.F32)
    with pytest.raises(S.SklError) as e:
        add(S.Vector(ctx, S.F32, 10).fill(1.0), S.Vector(ctx, S.F32, 11).fill(1.0))
    assert e.value.name == "SIZE_MISMATCH"
    with pytest.raises(S.SklError) as e:
        S.Map(ctx, A.NEG, S.F32, S.F32)(S.Vector(ctx, S.U8, 10).fill(1))
    assert e.value.name == "TYPE"
    _still_works(ctx)


def test_capture_rules():
    """several local devices capture into one graph; nested captures and host
    reads inside a capture are refused"""
    require_gpu()
    c2 = S.Context(2, devices=[0, 0])
    try:
        g = c2.capture(lambda: None)
        g.launch()
        g.destroy()
        v = S.Vector.from_numpy(c2, np.ones(100, np.float32)).set_distribution(S.BLOCK)
        w = S.Map(c2, A.NEG, S.F32, S.F32)(v)          # lives on the devices only
        with pytest.raises(S.SklError) as e:
            c2.capture(lambda: c2.capture(lambda: None))
        assert e.value.name == "INVALID_ARG"
        with pytest.raises(S.SklError) as e:
            c2.capture(lambda: w.to_numpy())
        assert e.value.name == "INVALID_ARG"
        assert np.array_equal(w.to_numpy(), -np.ones(100, np.float32))   # still usable
    finally:
        c2.finalize()
