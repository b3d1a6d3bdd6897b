"""The torch copies of the seeded generator (inputs.py, used for the 2^30 Scan
vectors) produce exactly the numpy streams (no GPU: torch on the CPU)."""
import numpy as np
import pytest
import torch

from paper_conf_pact_steuwerg13_b200 import inputs as I


@pytest.mark.parametrize("seed,start,n", [(4, 0, 5000), (4, (1 << 30) - 777, 777), (1, 123456789, 3001)])
def test_uniform_f32_torch_matches_numpy(seed, start, n):
    got = I.uniform_f32_torch(seed, n, device="cpu", start=start, chunk=1024).numpy()
    assert np.array_equal(got.view(np.uint32), I.uniform_f32(seed, n, start=start).view(np.uint32))


@pytest.mark.parametrize("seed,start,n,lo,hi", [(3, 0, 5000, -1000, 1000), (3, (1 << 30) - 999, 999, -1000, 1000),
                                                (5, 77, 4096, 0, 255), (9, 0, 2048, -2**30, 2**30 - 1)])
def test_uniform_int_torch_matches_numpy(seed, start, n, lo, hi):
    got = I.uniform_int_torch(seed, n, lo, hi, device="cpu", start=start, chunk=1000).numpy()
    assert np.array_equal(got, I.uniform_int(seed, n, lo, hi, np.int32, start=start))
