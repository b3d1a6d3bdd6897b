"""Pins for the CPU oracle (no GPU): the oracle checked against what the paper
and mathematics fix — hand-derived golden fixtures (tests/golden, each citing
its passage), closed forms, invariants, special cases that reduce to an
independent library routine (numpy / scipy), and brute force on tiny inputs.

Each pin is chosen so that a plausible slip in oracle.cpp (dropped term, wrong
sign or index, swapped operands, wrong boundary) fails at least one of them.
"""
import math

import numpy as np
import pytest
import scipy.ndimage as ndi

import oracle as O
from paper_conf_pact_steuwerg13_b200 import inputs as I
from conftest import read_golden


# ------------------------------------------------------------------ Map
def test_map_neg_flips_only_the_sign_bit():
    # P:L254 negation: IEEE negation flips bit 31 and nothing else, incl. +-0, inf, NaN
    x = np.array([0.0, -0.0, 1.5, -2.25, np.inf, -np.inf, np.nan, 1e-45, 3.4e38],
                 dtype=np.float32)
    x = np.concatenate([x, I.uniform_f32(11, 1000) - 0.5])
    y = O.map_(O.OM_NEG_F32, x)
    assert np.array_equal(y.view(np.uint32), x.view(np.uint32) ^ np.uint32(0x80000000))


def test_map_sqp1_is_two_separately_rounded_ops():
    # numpy fp32 evaluates x*x then +1 with two roundings (no FMA): independent twin.
    x = (I.uniform_f32(12, 4097) * 8 - 4).astype(np.float32)
    y = O.map_(O.OM_SQP1_F32, x)
    ref = (x * x).astype(np.float32) + np.float32(1.0)
    assert np.array_equal(y, ref)
    # and an FMA-contracted version differs somewhere (so the pin has teeth)
    fma = (x.astype(np.float64) * x.astype(np.float64) + 1.0).astype(np.float32)
    assert not np.array_equal(y, fma)


def test_map_int_wraps_mod_2_32():
    x = np.array([0, 1, -1, 2**31 - 1, -2**31, 715827882], dtype=np.int32)
    y = O.map_(O.OM_AFFINE_I32, x)
    ref = ((x.astype(np.int64) * 3 + 7) % 2**32).astype(np.uint32).view(np.int32)
    assert np.array_equal(y, ref)


def test_map_u8_invert_involution():
    x = np.arange(256, dtype=np.uint8)
    y = O.map_(O.OM_INV_U8, x)
    assert np.array_equal(y, x[::-1])
    assert np.array_equal(O.map_(O.OM_INV_U8, y), x)


# ------------------------------------------------------------------ Mandelbrot
def test_mandelbrot_golden_points():
    g = read_golden("mandelbrot_points.txt")[None]
    c = np.array([[r[0], r[1]] for r in g], dtype=np.float32)
    want = np.array([r[2] for r in g], dtype=np.uint32)
    got, tot = O.mandelbrot(c, 1000)
    assert np.array_equal(got, want)
    assert tot == int(want.sum())


def test_mandelbrot_grid_is_exact_and_minus2_pixel():
    g = I.mandel_grid(3072, 4096)
    # A22: both grid steps are 3*2^-12, so c is exact in fp32
    assert g[0, 1, 0] - g[0, 0, 0] == np.float32(3 * 2 ** -12)
    assert g[1, 0, 1] - g[0, 0, 1] == np.float32(3 * 2 ** -12)
    # c = -2 is pixel (row 1536, col 0): |z|^2 stays exactly 4 -> MAX (strict >)
    assert g[1536, 0, 0] == -2.0 and g[1536, 0, 1] == 0.0
    out, _ = O.mandelbrot(g[1536:1537, 0:1], 1000)
    assert out[0, 0] == 1000


def test_mandelbrot_escape_bound_and_symmetry():
    # |c| > 2 escapes after exactly one iteration (z1 = c); the set is symmetric
    # in conj(c) and the fp32 iteration is exactly symmetric in the sign of cy.
    rng_c = I.mandel_grid(96, 128)
    out, _ = O.mandelbrot(rng_c, 200)
    flipped = rng_c.copy()
    flipped[..., 1] = -flipped[..., 1]
    out2, _ = O.mandelbrot(flipped, 200)
    assert np.array_equal(out, out2)
    far = np.array([[2.5, 0], [0, -2.1], [-1.6, 1.6]], dtype=np.float32)
    o3, _ = O.mandelbrot(far, 1000)
    assert np.all(o3 == 1)


def test_mandelbrot_bruteforce_small_grid():
    # pure-Python fp32 (numpy scalar) loop on a tiny grid
    c = I.mandel_grid(12, 16)
    out, tot = O.mandelbrot(c, 60)
    f = np.float32
    for r in range(12):
        for k in range(16):
            cx, cy = c[r, k]
            x = y = f(0)
            n = 0
            while n < 60:
                xx, yy = f(x * x), f(y * y)
                if f(xx + yy) > f(4):
                    break
                y = f(f(f(2) * x) * y) + cy
                x = f(f(xx - yy) + cx)
                n += 1
            assert out[r, k] == n
    assert tot == int(out.sum())


# ------------------------------------------------------------------ Zip
def test_zip_add_mult_match_numpy_fp32():
    a = I.uniform_f32(1, 5000)
    b = I.uniform_f32(2, 5000)
    assert np.array_equal(O.zip_(O.OZ_ADD_F32, a, b), a + b)
    assert np.array_equal(O.zip_(O.OZ_MULT_F32, a, b), a * b)
    ai = I.uniform_int(3, 5000, -2**31, 2**31 - 1)
    bi = I.uniform_int(4, 5000, -2**31, 2**31 - 1)
    ref = ((ai.astype(np.int64) - bi.astype(np.int64)) % 2**32).astype(np.uint32).view(np.int32)
    assert np.array_equal(O.zip_(O.OZ_SUB_I32, ai, bi), ref)


def test_zip_size_mismatch_raises():
    with pytest.raises(ValueError):
        O.zip_(O.OZ_ADD_F32, np.zeros(3, np.float32), np.zeros(4, np.float32))


# ------------------------------------------------------------------ Reduce / Scan
def test_golden_scan_reduce():
    g = read_golden("scan_reduce_small.txt")
    x = np.array(g["input"][0], dtype=np.int32)
    assert np.array_equal(O.scan(O.OP_ADD_I32, x), np.array(g["scan"][0], dtype=np.int32))
    assert O.reduce_(O.OP_ADD_I32, x) == int(g["reduce"][0][0])


@pytest.mark.parametrize("n", [1, 2, 3, 31, 32, 33, 4097, 1 << 20])
def test_reduce_closed_forms(n):
    assert O.reduce_(O.OP_ADD_F32, np.ones(n, np.float32)) == float(n)
    idx = np.arange(n, dtype=np.int64)
    got = O.reduce_(O.OP_ADD_I32, (idx % 2**32).astype(np.uint32).view(np.int32))
    assert np.uint32(np.int32(got).view(np.uint32)) == np.uint32((n * (n - 1) // 2) % 2**32)


def test_reduce_empty_is_error():
    with pytest.raises(ValueError):
        O.reduce_(O.OP_ADD_F32, np.zeros(0, np.float32))


def test_reduce_order_pins_projections():
    # left projection -> v[0], right projection -> v[n-1]: a fold that reorders
    # or drops an operand fails one of these.
    x = I.uniform_f32(21, 777)
    assert O.reduce_(O.OP_LEFT_F32, x) == x[0]
    assert O.reduce_(O.OP_RIGHT_F32, x) == x[-1]
    assert O.reduce_(O.OP_MAX_F32, x) == x.max()


def _affine_apply(pairs, x):
    for a, b in pairs:
        x = (int(a) * x + int(b)) % 2**32
    return x


@pytest.mark.parametrize("n", [1, 2, 5, 64, 300])
def test_reduce_affine_equals_sequential_application(n):
    # non-commutative (+): composing maps must equal applying them in order
    p = I.uniform_int(22, 2 * n, 0, 2**32 - 1, np.uint64).astype(np.uint32).reshape(n, 2)
    a, b = O.reduce_(O.OP_AFFINE_U32, p)
    for x in (0, 1, 12345, 2**32 - 1):
        assert (int(a) * x + int(b)) % 2**32 == _affine_apply(p, x)


def test_scan_invariants():
    x = I.uniform_f32(23, 3000)
    s = O.scan(O.OP_ADD_F32, x)
    assert s[-1] == O.reduce_(O.OP_ADD_F32, x)
    assert np.array_equal(O.scan(O.OP_ADD_F32, np.ones(5000, np.float32)), np.arange(1, 5001))
    assert np.all(O.scan(O.OP_LEFT_F32, x) == x[0])
    assert np.array_equal(O.scan(O.OP_RIGHT_F32, x), x)
    # fp32 data, double accumulation: equals numpy's float64 cumsum up to rounding order
    assert np.allclose(s, np.cumsum(x.astype(np.float64)), rtol=1e-12)


def test_scan_bruteforce_definition():
    # out[i] = v1 (+) ... (+) v_{i+1}, recomputed from scratch per i
    n = 200
    p = I.uniform_int(24, 2 * n, 0, 2**32 - 1, np.uint64).astype(np.uint32).reshape(n, 2)
    s = O.scan(O.OP_AFFINE_U32, p)
    for i in (0, 1, 7, 63, 199):
        assert np.array_equal(s[i], O.reduce_(O.OP_AFFINE_U32, p[: i + 1]))
    xi = I.uniform_int(25, n, -1000, 1000)
    si = O.scan(O.OP_ADD_I32, xi)
    for i in range(n):
        assert si[i] == int(xi[: i + 1].astype(np.int64).sum())


def test_combine_gpu_order_and_exact_int_sum():
    G, n = 4, 1000
    r = I.uniform_int(26, G * n, -1000, 1000).reshape(G, n)
    assert np.array_equal(O.combine(O.OP_ADD_I32, r), r.astype(np.int64).sum(0).astype(np.int32))
    rf = I.uniform_f32(27, G * n).reshape(G, n)
    assert np.array_equal(O.combine(O.OP_LEFT_F32, rf), rf[0])
    assert np.array_equal(O.combine(O.OP_RIGHT_F32, rf), rf[-1])


# ------------------------------------------------------------------ MapOverlap
def test_golden_boxsum():
    g = read_golden("boxsum_4x4.txt")
    x = np.array(g["input"], dtype=np.float32)
    out = O.mapoverlap2d(O.OS_BOX3, x, 1, O.OB_NEUTRAL, 0.0)
    assert np.array_equal(out, np.array(g["output"], dtype=np.float32))


def test_golden_sobel_impulse():
    g = read_golden("sobel_impulse_5x5.txt")
    x = np.array(g["input"], dtype=np.uint8)
    out = O.mapoverlap2d(O.OS_SOBEL, x, 1, O.OB_NEUTRAL, 0)
    assert np.array_equal(out, np.array(g["output"], dtype=np.uint8))


def test_mapoverlap_identity_and_shift_orientation():
    x = I.image_f32(31, 37, 53)
    assert np.array_equal(O.mapoverlap2d(O.OS_IDENT, x, 1, O.OB_NEUTRAL, 0.0), x)
    # get(+1, 0): dx is the COLUMN offset (A15) -> left shift with neutral fill
    sx = O.mapoverlap2d(O.OS_SHIFT_X, x, 1, O.OB_NEUTRAL, 7.0)
    assert np.array_equal(sx[:, :-1], x[:, 1:]) and np.all(sx[:, -1] == 7.0)
    sy = O.mapoverlap2d(O.OS_SHIFT_Y, x, 1, O.OB_NEAREST, 0.0)
    assert np.array_equal(sy[:-1], x[1:]) and np.array_equal(sy[-1], x[-1])
    xu = I.image_u8(32, 9, 11)
    su = O.mapoverlap2d(O.OS_SHIFT_X, xu, 1, O.OB_NEAREST, 0)
    assert np.array_equal(su[:, :-1], xu[:, 1:]) and np.array_equal(su[:, -1], xu[:, -1])


@pytest.mark.parametrize("k", [1.0, 2.5])
def test_boxsum_constant_image(k):
    x = np.full((6, 7), k, np.float32)
    o = O.mapoverlap2d(O.OS_BOX3, x, 1, O.OB_NEUTRAL, 0.0)
    assert np.all(o[1:-1, 1:-1] == 9 * k)
    assert np.all(o[0, 1:-1] == 6 * k) and np.all(o[1:-1, 0] == 6 * k)
    assert o[0, 0] == 4 * k and o[-1, -1] == 4 * k
    on = O.mapoverlap2d(O.OS_BOX3, x, 1, O.OB_NEAREST, 0.0)
    assert np.all(on == 9 * k)


def test_boxsum_matches_scipy_correlate():
    x = I.image_f32(33, 40, 64)
    ref = ndi.correlate(x.astype(np.float64), np.ones((3, 3)), mode="constant", cval=0.0)
    o = O.mapoverlap2d(O.OS_BOX3, x, 1, O.OB_NEUTRAL, 0.0)
    assert np.allclose(o, ref, rtol=1e-6, atol=1e-6)
    refn = ndi.correlate(x.astype(np.float64), np.ones((3, 3)), mode="nearest")
    on = O.mapoverlap2d(O.OS_BOX3, x, 1, O.OB_NEAREST, 0.0)
    assert np.allclose(on, refn, rtol=1e-6, atol=1e-6)


def test_sobel_matches_scipy_and_ramp():
    x = I.image_u8(34, 45, 61)
    xi = x.astype(np.int64)
    kh = np.array([[-1, 0, 1], [-2, 0, 2], [-1, 0, 1]])   # rows = dy, cols = dx
    h = ndi.correlate(xi, kh, mode="constant", cval=0)
    v = ndi.correlate(xi, kh.T, mode="constant", cval=0)
    m = np.sqrt((h * h + v * v).astype(np.float32)).astype(np.int64)
    ref = np.minimum(m, 255).astype(np.uint8)
    assert np.array_equal(O.mapoverlap2d(O.OS_SOBEL, x, 1, O.OB_NEUTRAL, 0), ref)
    # horizontal ramp p = s*c: interior h = 8s, v = 0
    for s in (1, 5, 40):
        ramp = np.tile((np.arange(20) * s % 256).astype(np.uint8), (6, 1))
        o = O.mapoverlap2d(O.OS_SOBEL, ramp, 1, O.OB_NEUTRAL, 0)
        if 19 * s < 256:
            assert np.all(o[1:-1, 1:-1] == min(255, 8 * s))
    const = np.full((8, 8), 77, np.uint8)
    assert np.all(O.mapoverlap2d(O.OS_SOBEL, const, 1, O.OB_NEUTRAL, 0)[1:-1, 1:-1] == 0)


def test_gaussian_weights_and_impulse():
    w = O.gauss5_weights()
    # independent derivation: separable 1-D Gaussian outer product
    g1 = np.exp(-np.arange(-2, 3) ** 2 / 2.0)
    ref = np.outer(g1, g1) / np.outer(g1, g1).sum()
    assert np.array_equal(w, ref.astype(np.float32))
    assert abs(float(w.astype(np.float64).sum()) - 1.0) < 1e-6
    img = np.zeros((9, 9), np.float32)
    img[4, 4] = 1.0
    o = O.mapoverlap2d(O.OS_GAUSS5, img, 2, O.OB_NEUTRAL, 0.0)
    # impulse response = weight table, flipped (correlation) — symmetric here
    assert np.array_equal(o[2:7, 2:7], w[::-1, ::-1])
    assert np.count_nonzero(o) == 25


def test_gaussian_nearest_constant_and_scipy():
    x = np.full((7, 9), 0.7, np.float32)
    o = O.mapoverlap2d(O.OS_GAUSS5, x, 2, O.OB_NEAREST, 0.0)
    assert np.all(np.abs(o - np.float32(0.7)) <= 25 * np.spacing(np.float32(0.7)))
    y = I.image_f32(6, 30, 40)
    ref = ndi.correlate(y.astype(np.float64), O.gauss5_weights().astype(np.float64), mode="nearest")
    assert np.allclose(O.mapoverlap2d(O.OS_GAUSS5, y, 2, O.OB_NEAREST, 0.0), ref, rtol=0, atol=1e-6)


def test_mapoverlap1d_pins():
    v = I.uniform_f32(35, 100)
    assert np.array_equal(O.mapoverlap1d(O.OS_IDENT, v, 1, O.OB_NEUTRAL, 0.0), v)
    s = O.mapoverlap1d(O.OS_SHIFT_X, v, 1, O.OB_NEUTRAL, -1.0)
    assert np.array_equal(s[:-1], v[1:]) and s[-1] == -1.0
    b = O.mapoverlap1d(O.OS_BOX3, v, 1, O.OB_NEAREST, 0.0)
    ref = np.convolve(np.pad(v.astype(np.float64), 1, mode="edge"), np.ones(3), mode="valid")
    assert np.allclose(b, ref, rtol=1e-6)
    # 1-D is the matrix definition with a single row
    m = O.mapoverlap2d(O.OS_BOX3, v.reshape(1, -1), 1, O.OB_NEUTRAL, 0.0)
    assert np.array_equal(O.mapoverlap1d(O.OS_BOX3, v, 1, O.OB_NEUTRAL, 0.0), m[0])


# ------------------------------------------------------------------ Allpairs
def test_golden_allpairs():
    g = read_golden("allpairs_small.txt")
    a, b = np.array(g["A"], np.float32), np.array(g["B"], np.float32)
    assert np.array_equal(O.allpairs(O.AP_DOT, a, b), np.array(g["dot"], np.float32))
    assert np.array_equal(O.allpairs(O.AP_MANHATTAN, a, b), np.array(g["manhattan"], np.float32))


def test_allpairs_eq2_matrix_multiply_and_cityblock():
    from scipy.spatial.distance import cdist
    a = I.uniform_f32(71, 37 * 19).reshape(37, 19) - np.float32(0.5)
    bt = I.uniform_f32(72, 19 * 23).reshape(19, 23) - np.float32(0.5)   # B is d x m
    # Eq. (2): A x B = allpairs(dotProduct)(A, B^T)
    c64 = O.allpairs(O.AP_DOT_F64, a, np.ascontiguousarray(bt.T))
    assert np.allclose(c64, a.astype(np.float64) @ bt.astype(np.float64), rtol=1e-12, atol=1e-12)
    c32 = O.allpairs(O.AP_DOT, a, np.ascontiguousarray(bt.T))
    assert np.allclose(c32, c64, rtol=0, atol=19 * 2e-7)
    b = I.uniform_f32(73, 23 * 19).reshape(23, 19)
    man = O.allpairs(O.AP_MANHATTAN, a, b)
    assert np.allclose(man, cdist(a.astype(np.float64), b.astype(np.float64), "cityblock"), rtol=1e-6)
    # the fold is left to right in fp32: first column of a 1-column problem is |a-b|
    assert np.array_equal(O.allpairs(O.AP_MANHATTAN, a[:, :1], b[:, :1]), np.abs(a[:, :1] - b[:, :1].T))


# ------------------------------------------------------------------ Distributions
def test_golden_block_partition():
    for row in read_golden("block_partition.txt")[None]:
        n, G = int(row[0]), int(row[1])
        want = [(int(row[2 + 2 * g]), int(row[3 + 2 * g])) for g in range(G)]
        assert [O.block_range(n, G, g) for g in range(G)] == want


@pytest.mark.parametrize("n", [0, 1, 2, 7, 8, 9, 1000, 3072, 8193])
@pytest.mark.parametrize("G", [1, 2, 3, 4, 8])
def test_block_covers_once_in_order(n, G):
    parts = [O.block_range(n, G, g) for g in range(G)]
    cover = np.zeros(n, np.int64)
    prev_hi = 0
    for lo, hi in parts:
        assert lo == prev_hi and lo <= hi   # contiguous, disjoint, in GPU order
        cover[lo:hi] += 1
        prev_hi = hi
    assert prev_hi == n and np.all(cover == 1)


@pytest.mark.parametrize("d", [1, 2, 5])
def test_overlap_halo_is_neighbours_border(d):
    n, G = 50, 4
    for g in range(G):
        blo, bhi = O.block_range(n, G, g)
        lo, hi = O.overlap_range(n, G, g, d)
        assert lo == max(0, blo - d) and hi == min(n, bhi + d)
        if g > 0:  # top halo = last d units of the previous block
            plo, phi = O.block_range(n, G, g - 1)
            assert lo == max(plo, phi - d)


# ------------------------------------------------------------------ LM OSEM (W3, A29)
def _chord(p0, p1, N):
    """slab-clipping closed form of |segment ∩ [0,N]^3|"""
    p0, p1 = np.asarray(p0, np.float64), np.asarray(p1, np.float64)
    d = p1 - p0
    lo, hi = 0.0, 1.0
    for a in range(3):
        if d[a] == 0:
            if not (0 <= p0[a] <= N):
                return 0.0
            continue
        t0, t1 = (0 - p0[a]) / d[a], (N - p0[a]) / d[a]
        lo, hi = max(lo, min(t0, t1)), min(hi, max(t0, t1))
    return max(0.0, hi - lo) * float(np.linalg.norm(d))


def test_siddon_axis_aligned_row():
    N = 4
    vox, ln = O.siddon([-1, 1.5, 2.5], [N + 1, 1.5, 2.5], N)
    assert np.array_equal(vox, [(2 * N + 1) * N + x for x in range(N)])
    assert np.allclose(ln, 1.0)


def test_siddon_lengths_sum_to_chord_and_sample_bruteforce():
    N = 4
    ev = I.lmosem_events(I.SEED_LMOSEM, 10, N)
    for e in ev:
        vox, ln = O.siddon(e[:3], e[3:], N)
        assert abs(ln.sum() - _chord(e[:3], e[3:], N)) < 1e-9
        assert len(set(vox.tolist())) == len(vox)
        # brute force: dense sampling along the segment, per-voxel length
        t = (np.arange(200000) + 0.5) / 200000
        p = e[:3].astype(np.float64)[None] + t[:, None] * (e[3:] - e[:3]).astype(np.float64)[None]
        inside = np.all((p >= 0) & (p < N), axis=1)
        ijk = np.floor(p[inside]).astype(np.int64)
        lin = (ijk[:, 2] * N + ijk[:, 1]) * N + ijk[:, 0]
        L = float(np.linalg.norm((e[3:] - e[:3]).astype(np.float64)))
        ids, cnt = np.unique(lin, return_counts=True)
        bf = dict(zip(ids.tolist(), (cnt * L / 200000).tolist()))
        got = dict(zip(vox.tolist(), ln.tolist()))
        for k in set(bf) | set(got):
            assert abs(bf.get(k, 0.0) - got.get(k, 0.0)) < 2e-3 * L


def test_lmosem_invariants():
    N = 12
    ev = I.lmosem_events(I.SEED_LMOSEM, 3000, N)
    f = np.ones(N ** 3, np.float32)
    c, fnew, nhit, visits = O.lmosem(ev, N, f)
    # sum_v f[v] c[v] = #events with fp > 0 (exact in real arithmetic)
    assert abs(float((f.astype(np.float64) * c).sum()) - nhit) < 1e-6 * max(1, nhit)
    assert np.array_equal(fnew, f.astype(np.float64) * c)
    assert 0 < nhit <= 3000 and visits > nhit
    # with f = 1, fp_e = chord_e
    f2 = (1.0 + I.uniform_f32(8, N ** 3)).astype(np.float32)
    c2, _, nhit2, _ = O.lmosem(ev, N, f2)
    assert nhit2 == nhit
    assert abs(float((f2.astype(np.float64) * c2).sum()) - nhit2) < 1e-6 * nhit2


def test_lmosem_geometry_hit_rate():
    # A29 geometry: Monte-Carlo estimate in SURVEY §8(d): ~65.8% of events hit
    N = 30
    ev = I.lmosem_events(I.SEED_LMOSEM, 20000, N)
    _, _, nhit, _ = O.lmosem(ev, N, np.ones(N ** 3, np.float32))
    assert 0.60 < nhit / 20000 < 0.72


# ------------------------------------------------------------------ pins added in round 2
def test_row_sums_closed_forms_and_bruteforce():
    # constant-count matrix: every row sums to cols * k (closed form); counts near
    # 2^32 make the total overflow 32 bits, so a 32-bit accumulator fails
    for rows, cols, k in ((1, 1, 7), (3, 5, 1000), (4, 3, 2**32 - 1)):
        s = O.row_sums(np.full((rows, cols), k, np.uint32))
        assert s.dtype == np.uint64 and np.array_equal(s, np.full(rows, cols * k, np.uint64))
    # brute force (pure Python) on a random matrix, and a one-hot matrix that
    # catches a transposed index (row r holds its only non-zero in column r)
    c = I.uniform_int(41, 7 * 13, 0, 100000, np.uint64).astype(np.uint32).reshape(7, 13)
    s = O.row_sums(c)
    for r in range(7):
        assert int(s[r]) == sum(int(v) for v in c[r])
    eye = np.zeros((5, 9), np.uint32)
    for r in range(5):
        eye[r, r] = r + 1
    assert np.array_equal(O.row_sums(eye), np.arange(1, 6, dtype=np.uint64))
    # the Mandelbrot total equals the sum of its row sums
    counts, tot = O.mandelbrot(I.mandel_grid(24, 32), 300)
    assert int(O.row_sums(counts).sum()) == tot


def test_gaussian_weights_agree_with_the_user_program():
    # the user program (apps.gaussian5) and the oracle derive the W1
    # weights independently; they must agree bit for bit, and the %.9g literals
    # printed into the customising-function source must round-trip to them.
    import re
    from paper_conf_pact_steuwerg13_b200 import apps as A
    w = O.gauss5_weights()
    assert np.array_equal(A.gauss5_weights().view(np.uint32), w.view(np.uint32))
    lits = [np.float32(float(m)) for m in re.findall(r"acc \+ ([0-9.e+-]+)f \* get", A.gaussian5())]
    assert len(lits) == 25
    assert np.array_equal(np.array(lits, np.float32).view(np.uint32), w.reshape(-1).view(np.uint32))


@pytest.mark.parametrize("G", [1, 2, 3, 8])
def test_combine_affine_is_gpu_order_fold(G):
    # A25: replicas folded in GPU order 0..G-1 with a non-commutative operator
    n = 50
    p = I.uniform_int(42 + G, G * n * 2, 0, 2**32 - 1, np.uint64).astype(np.uint32).reshape(G, n, 2)
    out = O.combine(O.OP_AFFINE_U32, p)
    for i in (0, 17, n - 1):
        a, b = out[i]
        for x in (0, 3, 2**31 + 5):
            assert (int(a) * x + int(b)) % 2**32 == _affine_apply(p[:, i], x)
    # fp32 + accumulated in double: G ones -> G exactly
    assert np.all(O.combine(O.OP_ADD_F32, np.ones((G, n), np.float32)) == float(G))
