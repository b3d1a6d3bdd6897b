"""Host-side checks of the reasoning behind the tuned user functions in
paper_conf_pact_steuwerg13_b200/apps.py (no GPU; the GPU tests run the functions
themselves against the oracle)."""
import numpy as np

from paper_conf_pact_steuwerg13_b200 import apps as A


def test_sobel_tuned_root_margin():
    """apps.SOBEL_TUNED takes floor(sqrt.approx(min(m + 1/2, 65025.5))): for every
    m = h^2 + v^2 <= 2,080,800 the root of the clamped m + 1/2 has the same floor
    as sqrt(m) saturated at 255, and lies at least 0.00098 from every integer -
    far more than the estimate's error (relative ~2^-23, < 1e-4 here)"""
    m = np.arange(2_080_801, dtype=np.float64)
    k = np.minimum(m + 0.5, 65025.5)
    r = np.sqrt(k)
    assert np.array_equal(np.floor(r), np.minimum(np.floor(np.sqrt(m)), 255))
    dist = np.abs(r - np.round(r))
    assert dist.min() >= 0.00098
    assert (r.max() * 2.0 ** -22) < 1e-4        # the estimate's absolute error bound here
    # k is exact in fp32 (integer + 1/2 below 2^22), as the function forms it
    assert np.array_equal(k.astype(np.float32).astype(np.float64), k)


def test_sobel_tuned_difference_form_is_listing_1_5():
    """the regrouped h, v of apps.SOBEL_TUNED equal Listing 1.5's sums for every
    3x3 neighbourhood (integer identity, checked on random and extreme windows)"""
    rng = np.random.default_rng(5)
    g = rng.integers(0, 256, size=(20000, 3, 3)).astype(np.int64)
    g[:4] = [[[0] * 3] * 3, [[255] * 3] * 3, [[0, 0, 255]] * 3, [[255, 0, 0]] * 3]
    G = lambda dx, dy: g[:, dy + 1, dx + 1]  # noqa: E731  get(img, dx, dy)
    h_paper = -G(-1, -1) + G(1, -1) - 2 * G(-1, 0) + 2 * G(1, 0) - G(-1, 1) + G(1, 1)
    v_paper = -G(-1, -1) - 2 * G(0, -1) - G(1, -1) + G(-1, 1) + 2 * G(0, 1) + G(1, 1)
    h0, h1, h2 = G(1, -1) - G(-1, -1), G(1, 0) - G(-1, 0), G(1, 1) - G(-1, 1)
    v0, v1, v2 = G(-1, 1) - G(-1, -1), G(0, 1) - G(0, -1), G(1, 1) - G(1, -1)
    assert np.array_equal(h0 + 2 * h1 + h2, h_paper)
    assert np.array_equal(v0 + 2 * v1 + v2, v_paper)
    assert "int h = h0 + 2 * h1 + h2, v = v0 + 2 * v1 + v2;" in A.SOBEL_TUNED


def test_sobel_tuned_bias_addend_is_or():
    """apps.SOBEL_TUNED forms the biased m as h*h + (v*v + 0x4B000000): for every
    m <= 2 * 1020^2 the 32-bit sum has the bits of 0x4B000000 | m (m < 2^23), and
    that word read as fp32 is 2^23 + m exactly"""
    m = np.arange(2 * 1020 * 1020 + 1, dtype=np.uint32)
    biased = (m + np.uint32(0x4B000000)).astype(np.uint32)
    assert np.array_equal(biased, m | np.uint32(0x4B000000))
    assert np.array_equal(biased.view(np.float32).astype(np.float64), m.astype(np.float64) + 2.0 ** 23)
    assert "int m = h * h + (v * v + 0x4B000000);" in A.SOBEL_TUNED
