"""Multi-device tests on one GPU (logical-device mode): G logical
devices, each with its own stream and memory, exchanging data by device-to-device
copies.  Checks the distribution semantics (readings A1-A8, A25)
and that every skeleton's result is independent of G (bit-exact where the bar is
bit-exact)."""
import numpy as np
import pytest

import oracle as O
from gpu_util import rel_l2, require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu

GS = [2, 3, 4]


@pytest.fixture(scope="module", params=GS)
def ctx(request):
    require_gpu()
    c = S.Context(request.param, devices=[0] * request.param)
    yield c
    c.finalize()


def parts(c: S.Container, ctx):
    """per-device (first_unit, nunits) of the valid data"""
    return [c.local_part(g)[1:] for g in range(ctx.ndev)]


def test_block_copy_single_overlap_roundtrip(ctx):
    G = ctx.ndev
    x = I.uniform_f32(51, 1001)
    v = S.Vector.from_numpy(ctx, x)
    v.set_distribution(S.BLOCK)
    assert [p for p in parts(v, ctx)] == [(lo, hi - lo) for lo, hi in
                                          (O.block_range(1001, G, g) for g in range(G))]
    v.set_distribution(S.COPY)
    assert all(p == (0, 1001) for p in parts(v, ctx))
    v.set_distribution(S.SINGLE, G - 1)
    assert parts(v, ctx)[G - 1] == (0, 1001) and all(p == (0, 0) for p in parts(v, ctx)[:-1])
    v.set_distribution(S.OVERLAP, 3)
    for g in range(G):
        lo, hi = O.overlap_range(1001, G, g, 3)
        assert parts(v, ctx)[g] == (lo, hi - lo)
    v.set_distribution(S.BLOCK)
    assert np.array_equal(v.to_numpy(), x)


def test_matrix_overlap_halo_equals_neighbour_rows(ctx):
    G = ctx.ndev
    x = I.image_f32(52, 50, 33)
    m = S.Matrix.from_numpy(ctx, x).set_distribution(S.BLOCK)
    m.set_distribution(S.OVERLAP, 2)
    import ctypes
    for g in range(G):
        ptr, first, n = m.local_part(g)
        lo, hi = O.overlap_range(50, G, g, 2)
        assert (first, n) == (lo, hi - lo)
        # borrowed device pointer: read it through torch (CUDA array interface, zero copy)
        import torch

        class View:
            __cuda_array_interface__ = {"shape": (n, 33), "typestr": "<f4", "data": (ptr, False),
                                        "version": 3, "strides": None}
        ctx.sync()
        host = torch.as_tensor(View(), device="cuda").cpu().numpy()
        assert np.array_equal(host, x[lo:hi])


@pytest.mark.parametrize("n", [7, 1000, 100003])
def test_map_zip_independent_of_G(ctx, n):
    x, y = I.uniform_f32(53, n), I.uniform_f32(54, n)
    neg = S.Map(ctx, A.SQP1, S.F32, S.F32)
    mult = S.Zip(ctx, A.MULT, S.F32, S.F32, S.F32)
    vx = S.Vector.from_numpy(ctx, x).set_distribution(S.BLOCK)
    vy = S.Vector.from_numpy(ctx, y).set_distribution(S.COPY)   # A7: right follows left
    assert np.array_equal(neg(vx).to_numpy(), O.map_(O.OM_SQP1_F32, x))
    r = mult(vx, vy)
    assert r.distribution()[0] == S.BLOCK
    assert np.array_equal(r.to_numpy(), O.zip_(O.OZ_MULT_F32, x, y))
    # copy input: every device computes everything (A8)
    vc = S.Vector.from_numpy(ctx, x).set_distribution(S.COPY)
    rc = neg(vc)
    assert rc.distribution()[0] == S.COPY and np.array_equal(rc.to_numpy(), O.map_(O.OM_SQP1_F32, x))


@pytest.mark.parametrize("n", [5, 4097, 300001])
def test_reduce_cross_device_ordered(ctx, n):
    aff = ctx.struct_type("Aff", A.AFFINE_DECL, 8, 4)
    red = S.Reduce(ctx, A.AFFINE_COMPOSE, aff)
    p = I.uniform_int(55, 2 * n, 0, 2**32 - 1, np.uint64).astype(np.uint32).reshape(n, 2)
    v = S.Vector(ctx, aff, n).copy_in(p)
    v.set_distribution(S.BLOCK)
    assert np.array_equal(red(v).scalar(np.uint32), O.reduce_(O.OP_AFFINE_U32, p))
    s = S.Reduce(ctx, A.SUM, S.F32)
    x = I.uniform_f32(56, n)
    got = float(s(S.Vector.from_numpy(ctx, x).set_distribution(S.BLOCK)).scalar())
    ref = O.reduce_(O.OP_ADD_F32, x)
    assert abs(got - ref) <= 1e-5 * abs(ref)
    left = S.Reduce(ctx, A.LEFT_F32, S.F32)
    right = S.Reduce(ctx, A.RIGHT_F32, S.F32)
    vx = S.Vector.from_numpy(ctx, x).set_distribution(S.BLOCK)
    assert left(vx).scalar() == x[0] and right(vx).scalar() == x[-1]


@pytest.mark.parametrize("n", [3, 8193, 200001])
def test_scan_carry_in(ctx, n):
    aff = ctx.struct_type("Aff", A.AFFINE_DECL, 8, 4)
    sa = S.Scan(ctx, A.AFFINE_COMPOSE, aff)
    p = I.uniform_int(57, 2 * n, 0, 2**32 - 1, np.uint64).astype(np.uint32).reshape(n, 2)
    v = S.Vector(ctx, aff, n).copy_in(p).set_distribution(S.BLOCK)
    got = sa(v).to_numpy(np.uint32).reshape(n, 2)
    assert np.array_equal(got, O.scan(O.OP_AFFINE_U32, p))
    si = S.Scan(ctx, A.ADD_I32, S.I32)
    xi = I.uniform_int(58, n, -1000, 1000)
    assert np.array_equal(si(S.Vector.from_numpy(ctx, xi).set_distribution(S.BLOCK)).to_numpy(),
                          O.scan(O.OP_ADD_I32, xi))
    sf = S.Scan(ctx, A.ADD, S.F32)
    x = I.uniform_f32(59, n)
    assert rel_l2(sf(S.Vector.from_numpy(ctx, x).set_distribution(S.BLOCK)).to_numpy(),
                  O.scan(O.OP_ADD_F32, x)) <= 1e-5


@pytest.mark.parametrize("shape", [(5, 9), (64, 200), (301, 257)])
def test_mapoverlap_halo_exchange(ctx, shape):
    sob = S.MapOverlap(ctx, A.SOBEL, S.U8, S.U8, 1, S.NEUTRAL, 0)
    gau = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
    xu = I.image_u8(I.SEED_SOBEL, *shape)
    assert np.array_equal(sob(S.Matrix.from_numpy(ctx, xu)).to_numpy(),
                          O.mapoverlap2d(O.OS_SOBEL, xu, 1, O.OB_NEUTRAL, 0))
    xf = I.image_f32(I.SEED_GAUSS, *shape)
    m = S.Matrix.from_numpy(ctx, xf)
    a = gau(m)
    assert a.distribution()[0] == S.BLOCK
    b = gau(a)  # block output -> overlap(2): halo refresh only
    r1 = O.mapoverlap2d(O.OS_GAUSS5, xf, 2, O.OB_NEAREST, 0.0)
    assert np.array_equal(a.to_numpy(), r1)
    assert np.array_equal(b.to_numpy(), O.mapoverlap2d(O.OS_GAUSS5, r1, 2, O.OB_NEAREST, 0.0))


def test_copy_combine_to_block(ctx):
    """copy(+) -> block (A25): every device adds its own events into its replica;
    leaving copy folds the replicas in GPU order."""
    G = ctx.ndev
    n, m = 5000, 97
    idx = I.uniform_int(60, n, 0, m - 1)
    w = I.uniform_int(61, n, -50, 50)
    ev2 = ctx.struct_type("Ev2", "struct Ev2 { int v, w; };", 8, 4)
    hist = S.Map(ctx, "void h(Ev2 e, int* c){ atomicAdd(&c[e.v], e.w); }", ev2, S.VOID,
                 extra=[S.I32 | S.PTR])
    ev = S.Vector(ctx, ev2, n).copy_in(np.stack([idx, w], 1).astype(np.int32))
    ev.set_distribution(S.BLOCK)
    addi = S.Reduce(ctx, A.ADD_I32, S.I32)
    c = S.Vector(ctx, S.I32, m).set_distribution(S.COPY, 0, addi)
    c.fill(0)
    hist(ev, (c, S.WRITE))
    # oracle: per-device replicas (block of events g into replica g), folded in GPU order
    reps = np.zeros((G, m), np.int32)
    for g in range(G):
        lo, hi = O.block_range(n, G, g)
        np.add.at(reps[g], idx[lo:hi], w[lo:hi])
    want = O.combine(O.OP_ADD_I32, reps)
    c.set_distribution(S.BLOCK)
    assert np.array_equal(c.to_numpy(), want)
    # and copy(+) -> copy leaves identical replicas
    c2 = S.Vector(ctx, S.I32, m).set_distribution(S.COPY, 0, addi)
    c2.fill(0)
    hist(ev, (c2, S.WRITE))
    c2.set_distribution(S.COPY, 0, addi)
    assert np.array_equal(c2.to_numpy(), want)


def test_lmosem_subset_small(ctx):
    N, nev = 16, 20000
    evd = ctx.struct_type("Event", A.EVENT_DECL, A.EVENT_SIZE, 4)
    lm = S.Map(ctx, A.lmosem_map(N), evd, S.VOID, extra=[S.F32 | S.PTR, S.F32 | S.PTR])
    upd = S.Zip(ctx, A.LMOSEM_UPDATE, S.F32, S.F32, S.F32)
    addf = S.Reduce(ctx, A.ADD, S.F32)
    events = I.lmosem_events(I.SEED_LMOSEM, nev, N)
    f0 = (1.0 + 0.5 * I.uniform_f32(8, N ** 3)).astype(np.float32)
    ev = S.Vector(ctx, evd, nev).copy_in(events).set_distribution(S.BLOCK)
    f = S.Vector.from_numpy(ctx, f0).set_distribution(S.COPY)
    c = S.Vector(ctx, S.F32, N ** 3).set_distribution(S.COPY, 0, addf)
    c.fill(0.0)
    lm(ev, f, (c, S.WRITE))
    c.set_distribution(S.BLOCK)              # copy(+) -> block combine
    f.set_distribution(S.BLOCK)
    fn = upd(f, c)
    c_ref, fn_ref, nhit, _ = O.lmosem(events, N, f0)
    assert rel_l2(c.to_numpy(), c_ref) <= 1e-4
    assert rel_l2(fn.to_numpy(), fn_ref) <= 1e-4
    # invariant: sum f*c = #events with fp > 0
    assert abs(float(np.dot(f0.astype(np.float64), c.to_numpy().astype(np.float64))) - nhit) <= 1e-3 * nhit


@pytest.mark.parametrize("n", [5, 4099, (1 << 20) + 7])
def test_reduce_of_unaligned_parts(ctx, n):
    """after overlap(1) -> block the parts keep their halo room, so device g's
    first element sits 4 bytes into its buffer: Reduce takes the unaligned
    (scalar) kernel, fused or not (found by tests/test_gpu_fuzz.py)"""
    x = I.uniform_f32(63, n) - np.float32(0.25)
    v = S.Vector.from_numpy(ctx, x).set_distribution(S.OVERLAP, 1)
    v.set_distribution(S.BLOCK)
    red = S.Reduce(ctx, A.SUM, S.F32)
    ref = O.reduce_(O.OP_ADD_F32, x)
    scale = float(np.abs(x).sum())
    assert abs(float(red(v).scalar()) - ref) <= 1e-5 * scale
    add = S.Zip(ctx, A.ADD, S.F32, S.F32, S.F32)
    ref2 = O.reduce_(O.OP_ADD_F32, O.zip_(O.OZ_ADD_F32, x, x))
    assert abs(float(red(add(v, v)).scalar()) - ref2) <= 1e-5 * 2 * scale
    right = S.Reduce(ctx, A.RIGHT_F32, S.F32)
    assert right(v).scalar() == x[-1]
