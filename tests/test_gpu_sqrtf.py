"""sqrtf inside a customising function (prelude.cuh skl_sqrtf): IEEE-754
correctly rounded for every one of the 2^32 fp32 inputs, i.e. bit for bit what
the library's -prec-sqrt=true contract (and the oracle's C sqrtf, e.g. in
Listing 1.5's (int)sqrtf((float)(h*h + v*v))) promises.  Reference:
numpy's fp32 square root (correctly rounded, denormals kept); NaN inputs and
negative inputs must give NaN, +-0 and +inf themselves."""
import numpy as np
import pytest

from gpu_util import require_gpu
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu

SQRT_F32 = "float rt(float x){ return sqrtf(x); }"


def test_sqrtf_all_2_32_inputs():
    require_gpu()
    c = S.Context(1)
    try:
        m = S.Map(c, SQRT_F32, S.F32, S.F32)
        chunk = 1 << 27
        for start in range(0, 1 << 32, chunk):
            bits = np.arange(start, start + chunk, dtype=np.uint64).astype(np.uint32)
            x = bits.view(np.float32)
            got = m(S.Vector.from_numpy(c, x)).to_numpy()
            with np.errstate(invalid="ignore"):
                ref = np.sqrt(x)
            nan = np.isnan(ref)
            assert np.array_equal(np.isnan(got), nan), hex(start)
            assert np.array_equal(got.view(np.uint32)[~nan], ref.view(np.uint32)[~nan]), hex(start)
    finally:
        c.finalize()


def test_sqrtf_special_values():
    require_gpu()
    c = S.Context(1)
    try:
        m = S.Map(c, SQRT_F32, S.F32, S.F32)
        x = np.array([0.0, -0.0, np.inf, -np.inf, np.nan, -1.0, 1.0, 4.0, 2.0 ** -149, 2.0 ** -126,
                      2.0 ** -101, np.nextafter(np.float32(2.0 ** -101), np.float32(0)),
                      np.finfo(np.float32).max, 65025.0, 65024.0], dtype=np.float32)
        got = m(S.Vector.from_numpy(c, x)).to_numpy()
        assert got[0] == 0.0 and not np.signbit(got[0])
        assert got[1] == 0.0 and np.signbit(got[1])
        assert got[2] == np.inf
        assert np.isnan(got[3]) and np.isnan(got[4]) and np.isnan(got[5])
        assert got[6] == 1.0 and got[7] == 2.0
        assert got[8] == np.sqrt(x[8]) and got[9] == np.float32(2.0 ** -63)
        with np.errstate(invalid="ignore"):
            assert np.array_equal(got[10:].view(np.uint32), np.sqrt(x[10:]).view(np.uint32))
    finally:
        c.finalize()
