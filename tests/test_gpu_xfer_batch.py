"""Batched transfer kernel (builtin.cu skl_xfer_batch): with
several logical devices in one process every redistribution move into a GPU
runs as one kernel launch, copying each segment in 16/8/4/1-byte units by the
common alignment of its source and destination, with bytewise heads and tails.
Every replica / part / halo is read back through its borrowed device pointer
and compared with the host array (P:L205-231 distributions), for element sizes
and lengths that give every misalignment; and the result is identical with the
kernel switched off (copy engines)."""
import numpy as np
import pytest

import oracle as O
from gpu_util import require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu


def device_bytes(ptr: int, nbytes: int) -> np.ndarray:
    import torch

    class View:
        __cuda_array_interface__ = {"shape": (nbytes,), "typestr": "|u1", "data": (ptr, False), "version": 3,
                                    "strides": None}
    return torch.as_tensor(View(), device="cuda").cpu().numpy()


def check_parts(ctx, c: S.Container, host: np.ndarray, unit_bytes: int):
    """every device's valid units equal the host array's units"""
    ctx.sync()
    hb = host.view(np.uint8).reshape(-1)
    for g in range(ctx.ndev):
        ptr, first, n = c.local_part(g)
        if n == 0:
            continue
        got = device_bytes(ptr, n * unit_bytes)
        assert np.array_equal(got, hb[first * unit_bytes:(first + n) * unit_bytes]), f"device {g}"


CASES = [(np.uint8, S.U8), (np.int32, S.I32), (np.float64, S.F64)]


@pytest.mark.parametrize("G", [2, 3, 5])
@pytest.mark.parametrize("n", [1, 17, 1001, 65537, 1 << 20])
@pytest.mark.parametrize("dt,st", CASES)
def test_vector_redistributions_bytewise(G, n, dt, st):
    require_gpu()
    ctx = S.Context(G, devices=[0] * G)
    try:
        x = (I.uniform_int(61, n, 0, 255, dtype=np.int64) * 7 + 3).astype(dt)
        v = S.Vector.from_numpy(ctx, x, st)
        ub = x.itemsize
        for kind, arg in ((S.BLOCK, 0), (S.COPY, 0), (S.SINGLE, G - 1), (S.BLOCK, 0), (S.OVERLAP, 3),
                          (S.SINGLE, 0), (S.COPY, 0), (S.OVERLAP, 1), (S.BLOCK, 0)):
            v.set_distribution(kind, arg)
            check_parts(ctx, v, x, ub)
        assert np.array_equal(v.to_numpy(), x)
    finally:
        ctx.finalize()


@pytest.mark.parametrize("G", [2, 4])
@pytest.mark.parametrize("rows,cols", [(37, 13), (64, 1024), (101, 3)])
def test_matrix_halo_refresh_after_stencil(G, rows, cols):
    """overlap(2) halos refreshed after a stencil wrote the block parts (the
    MapOverlap output keeps spare halo room, so only 2 rows per boundary move)"""
    require_gpu()
    ctx = S.Context(G, devices=[0] * G)
    try:
        ctx.set_option("halo_push", 0)
        x = I.image_f32(62, rows, cols)
        m = S.Matrix.from_numpy(ctx, x)
        ident = S.MapOverlap(ctx, A.IDENT2D, S.F32, S.F32, 2, S.NEAREST, 0.0)
        out = ident(m)
        out.set_distribution(S.OVERLAP, 2)
        check_parts(ctx, out, x, cols * 4)
        ref = O.mapoverlap2d(O.OS_GAUSS5, x, 2, O.OB_NEAREST, 0.0)
        gau = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
        assert np.array_equal(gau(out).to_numpy(), ref)
    finally:
        ctx.finalize()


@pytest.mark.parametrize("G", [2, 3, 4])
def test_copy_combine_kernel_vs_copy_engines(G):
    """copy(+) -> block of replicas that all differ, with the batched kernel and
    with cudaMemcpy: the same bits, equal to the GPU-order fold (A25)"""
    require_gpu()
    n = 150 ** 3
    res = []
    for xk in (1, 0):
        ctx = S.Context(G, devices=[0] * G)
        try:
            ctx.set_option("xfer_kernel", xk)
            add = S.Reduce(ctx, A.ADD, S.F32)
            c = S.Vector(ctx, S.F32, n).set_distribution(S.COPY, 0, add)
            c.fill(0.0)
            # every device adds its own pattern over the whole replica (a copy
            # input is computed whole on each device, A8)
            idx = S.Vector.from_numpy(ctx, np.arange(n, dtype=np.int32)).set_distribution(S.COPY)
            touch = S.Map(ctx, "void t(int i, float* c) { c[i] = c[i] + 0.25f * (float)(i % 7) + 1.0f; }",
                          S.I32, S.VOID, extra=[S.F32 | S.PTR])
            touch(idx, (c, S.WRITE))
            c.set_distribution(S.BLOCK)
            res.append(c.to_numpy())
        finally:
            ctx.finalize()
    i = np.arange(n)
    one = (np.float32(0.25) * (i % 7).astype(np.float32) + np.float32(1.0)).astype(np.float32)
    ref = one.copy()
    for _ in range(G - 1):
        ref = (ref + one).astype(np.float32)
    assert np.array_equal(res[0], res[1])
    assert np.array_equal(res[0], ref)
