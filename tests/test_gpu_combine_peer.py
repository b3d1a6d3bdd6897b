"""copy(+) -> block fused with its exchange (combine_peer): with
one process driving every device, device g folds its block slice straight out
of every replica in device order and writes it in place into its own replica.
Checked against the oracle's GPU-order fold (reading A25) with a
non-commutative operator (affine composition, so a wrong replica order fails),
integer and fp32 adds, matrices (row units), slices that are not 16-byte
aligned, and against the staged path (combine_peer=0)."""
import numpy as np
import pytest

import oracle as O
from gpu_util import require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module", params=[2, 3, 4, 8])
def ctx(request):
    require_gpu()
    G = request.param
    c = S.Context(G, devices=[0] * G)
    yield c
    c.finalize()


def diverged_replicas(ctx, m, seed):
    """an Aff copy(compose) Vector whose replica g holds its own values at every
    position: a void Map over G*m block-distributed events (device g gets events
    g*m .. g*m+m-1, event k writes position k % m)"""
    G = ctx.ndev
    aff = ctx.struct_type("Aff", A.AFFINE_DECL, 8, 4)
    ev3 = ctx.struct_type("Ev3", "struct Ev3 { unsigned int i, a, b; };", 12, 4)
    put = S.Map(ctx, "void put(Ev3 e, Aff* c){ Aff v; v.a = e.a; v.b = e.b; c[e.i] = v; }", ev3, S.VOID,
                extra=[aff | S.PTR])
    comp = S.Reduce(ctx, A.AFFINE_COMPOSE, aff)
    n = G * m
    ab = I.uniform_int(seed, 2 * n, 0, 2 ** 32 - 1, np.uint64).astype(np.uint32).reshape(n, 2)
    evs = np.zeros((n, 3), np.uint32)
    evs[:, 0] = np.arange(n) % m
    evs[:, 1:] = ab
    ev = S.Vector(ctx, ev3, n).copy_in(evs).set_distribution(S.BLOCK)
    c = S.Vector(ctx, aff, m).set_distribution(S.COPY, 0, comp)
    put(ev, (c, S.WRITE))
    reps = ab.reshape(G, m, 2)
    return c, reps, (ev, put, comp)


@pytest.mark.parametrize("m", [1, 7, 1000, 4099, 100003])
def test_noncommutative_fold_order(ctx, m):
    c, reps, keep = diverged_replicas(ctx, m, 70 + m % 13)
    before = ctx.counter("launches")
    c.set_distribution(S.BLOCK)
    got = c.to_numpy(np.uint32).reshape(m, 2)
    assert np.array_equal(got, O.combine(O.OP_AFFINE_U32, reps))
    assert ctx.counter("launches") > before


def test_paths_bitexact_and_oracle_f32(ctx):
    """fp32 (+): the staged path (0), the one-launch fused path (1) and the
    per-device fused kernels (2) all fold in GPU order, so they agree bit for
    bit; against the oracle's double fold within the fp32 tolerance (A30)"""
    G = ctx.ndev
    m = 3 * 5003 + 1
    add = S.Reduce(ctx, A.ADD, S.F32)
    x = I.uniform_f32(75, G * m) - np.float32(0.5)
    ev2 = ctx.struct_type("EvF", "struct EvF { unsigned int i; float w; };", 8, 4)
    put = S.Map(ctx, "void putf(EvF e, float* c){ c[e.i] = e.w; }", ev2, S.VOID, extra=[S.F32 | S.PTR])
    evs = np.zeros(G * m, dtype=[("i", np.uint32), ("w", np.float32)])
    evs["i"] = np.arange(G * m) % m
    evs["w"] = x
    ev = S.Vector(ctx, ev2, G * m).copy_in(evs.view(np.uint8)).set_distribution(S.BLOCK)
    got = []
    try:
        for peer in (0, 1, 2):
            ctx.set_option("combine_peer", peer)
            c = S.Vector(ctx, S.F32, m).set_distribution(S.COPY, 0, add)
            put(ev, (c, S.WRITE))
            c.set_distribution(S.BLOCK)
            got.append(c.to_numpy())
    finally:
        ctx.set_option("combine_peer", 1)
    assert np.array_equal(got[0], got[1]) and np.array_equal(got[0], got[2])
    ref = O.combine(O.OP_ADD_F32, x.reshape(G, m))
    assert np.max(np.abs(got[1] - ref)) <= 1e-6 * np.max(np.abs(x)) * G


@pytest.mark.parametrize("peer", [1, 2])
def test_per_device_kernels_order(ctx, peer):
    """the per-device kernels (combine_peer=2) and the one-launch kernel keep the
    GPU order for a non-commutative operator"""
    ctx.set_option("combine_peer", peer)
    try:
        c, reps, keep = diverged_replicas(ctx, 5003, 79)
        c.set_distribution(S.BLOCK)
        assert np.array_equal(c.to_numpy(np.uint32).reshape(5003, 2), O.combine(O.OP_AFFINE_U32, reps))
    finally:
        ctx.set_option("combine_peer", 1)


@pytest.mark.parametrize("peer", [0, 1, 2])
def test_matrix_rows_and_unaligned_slices(ctx, peer):
    """a Matrix combines by rows; 13-column int32 rows put the block slices at
    offsets that are not 16-byte aligned (scalar kernel path)"""
    G = ctx.ndev
    ctx.set_option("combine_peer", peer)
    R, C = 37, 13
    addi = S.Reduce(ctx, A.ADD_I32, S.I32)
    vals = I.uniform_int(77, G * R * C, -1000, 1000).astype(np.int32)
    ev2 = ctx.struct_type("EvI", "struct EvI { int i, w; };", 8, 4)
    put = S.Map(ctx, "void puti(EvI e, int* c){ c[e.i] = e.w; }", ev2, S.VOID, extra=[S.I32 | S.PTR])
    evs = np.stack([np.arange(G * R * C) % (R * C), vals], 1).astype(np.int32)
    ev = S.Vector(ctx, ev2, G * R * C).copy_in(evs).set_distribution(S.BLOCK)
    c = S.Matrix(ctx, S.I32, R, C).set_distribution(S.COPY, 0, addi)
    put(ev, (c, S.WRITE))
    c.set_distribution(S.BLOCK)
    want = O.combine(O.OP_ADD_I32, vals.reshape(G, R * C)).reshape(R, C)
    assert np.array_equal(c.to_numpy(), want)
    # the folded container is usable as a block input (e.g. a Map) afterwards
    neg = S.Map(ctx, "int ng(int x){ return -x; }", S.I32, S.I32)
    assert np.array_equal(neg(c).to_numpy(), -want)
    ctx.set_option("combine_peer", 1)
