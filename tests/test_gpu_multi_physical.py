"""Multi-GPU paths across PHYSICAL devices: run when the box has
at least 2 GPUs, skipped otherwise (the round's GPU calls have one).

* one process driving 2..N GPUs: peer access to the peers' stream-ordered pools,
  the batched pull kernel for every redistribution, the fused halo push of an
  iterated stencil, the fused copy(+) -> block fold and the cross-device Reduce
  fold, each against the oracle;
* one process per GPU over the IPC transport (2 ranks on GPUs 0 and 1).
"""
import multiprocessing as mp
import os
import sys

import numpy as np
import pytest

import oracle as O
from gpu_util import require_gpu
from paper_conf_pact_steuwerg13_b200 import apps as A
from paper_conf_pact_steuwerg13_b200 import inputs as I
from paper_conf_pact_steuwerg13_b200 import skl as S

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def ngpus():
    require_gpu()
    import torch
    return torch.cuda.device_count()


@pytest.fixture(params=[2, 4, 8])
def phys_ctx(request):
    n = request.param
    if ngpus() < n:
        pytest.skip(f"needs {n} GPUs")
    c = S.Context(n, devices=list(range(n)))
    yield c
    c.finalize()


def test_redistributions_across_gpus(phys_ctx):
    c = phys_ctx
    x = I.uniform_f32(1, 1000003)
    v = S.Vector.from_numpy(c, x)
    for d, arg in ((S.BLOCK, 0), (S.COPY, 0), (S.SINGLE, c.ndev - 1), (S.OVERLAP, 7), (S.BLOCK, 0)):
        v.set_distribution(d, arg)
        assert np.array_equal(v.to_numpy(), x), (d, arg)
    assert c.counter("p2p_bytes") > 0


def test_reduce_and_scan_across_gpus(phys_ctx):
    c = phys_ctx
    x = I.uniform_f32(2, 777777)
    vx = S.Vector.from_numpy(c, x).set_distribution(S.BLOCK)
    assert S.Reduce(c, A.RIGHT_F32, S.F32)(vx).scalar() == x[-1]
    assert S.Reduce(c, A.LEFT_F32, S.F32)(vx).scalar() == x[0]
    xi = I.uniform_int(3, 777777, -1000, 1000)
    out = S.Scan(c, A.ADD_I32, S.I32)(S.Vector.from_numpy(c, xi).set_distribution(S.BLOCK))
    assert np.array_equal(out.to_numpy(), O.scan(O.OP_ADD_I32, xi))


def test_iterated_stencil_halo_push_across_gpus(phys_ctx):
    c = phys_ctx
    img = I.image_f32(I.SEED_GAUSS, 1024, 512)
    gau = S.MapOverlap(c, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
    a = S.Matrix.from_numpy(c, img)
    b = gau(a)
    t = gau(b)
    b = gau(t, out=b)
    ref = img
    for _ in range(3):
        ref = O.mapoverlap2d(O.OS_GAUSS5, ref, 2, O.OB_NEAREST, 0.0)
    assert np.array_equal(b.to_numpy(), ref)
    assert c.counter("halo_push_bytes") > 0


def test_graph_of_iterated_stencil_across_gpus(phys_ctx):
    """the iterated stencil recorded as one multi-device CUDA graph (kernels and
    halo pushes on every GPU) and replayed"""
    c = phys_ctx
    img = I.image_f32(I.SEED_GAUSS + 1, 1024, 512)
    gau = S.MapOverlap(c, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
    a = S.Matrix.from_numpy(c, img)
    b = S.Matrix(c, S.F32, 1024, 512)
    t = S.Matrix(c, S.F32, 1024, 512)

    def it():
        gau(a, out=b)
        gau(b, out=t)
        gau(t, out=b)

    it()
    g = c.capture(it)
    b.fill(0.0)
    g.launch()
    ref = img
    for _ in range(3):
        ref = O.mapoverlap2d(O.OS_GAUSS5, ref, 2, O.OB_NEAREST, 0.0)
    assert np.array_equal(b.to_numpy(), ref)
    g.destroy()


def test_copy_add_to_block_across_gpus(phys_ctx):
    c = phys_ctx
    n = 150 ** 3
    addf = S.Reduce(c, A.ADD, S.F32)
    cv = S.Vector(c, S.F32, n).set_distribution(S.COPY, 0, addf).fill(0.0)
    idx = S.Vector.from_numpy(c, np.arange(n, dtype=np.int32)).set_distribution(S.BLOCK)
    touch = S.Map(c, "void touch(int i, float* c) { c[i] = 1.0f + (float)(i % 3); }", S.I32, S.VOID,
                  extra=[S.F32 | S.PTR])
    touch(idx, (cv, S.WRITE))
    cv.set_distribution(S.BLOCK)
    assert np.array_equal(cv.to_numpy(), (1.0 + (np.arange(n) % 3)).astype(np.float32))


def _ipc_worker(rank, world, nid, q):
    try:
        os.environ["SKL_COMM"] = "ipc"
        sys.path.insert(0, ROOT)
        import oracle as O2
        from paper_conf_pact_steuwerg13_b200 import apps as A2
        from paper_conf_pact_steuwerg13_b200 import inputs as I2
        from paper_conf_pact_steuwerg13_b200 import skl as S2
        ctx = S2.Context.dist(rank, world, rank, nid)
        img = I2.image_u8(I2.SEED_SOBEL, 301, 272)
        sob = S2.MapOverlap(ctx, A2.SOBEL_TUNED, S2.U8, S2.U8, 1, S2.NEUTRAL, 0)
        b = sob(sob(S2.Matrix.from_numpy(ctx, img)))
        ref = O2.mapoverlap2d(O2.OS_SOBEL, O2.mapoverlap2d(O2.OS_SOBEL, img, 1, O2.OB_NEUTRAL, 0), 1,
                              O2.OB_NEUTRAL, 0)
        assert np.array_equal(b.to_numpy(), ref)
        xi = I2.uniform_int(3, 100003, -1000, 1000)
        assert np.array_equal(S2.Scan(ctx, A2.ADD_I32, S2.I32)(S2.Vector.from_numpy(ctx, xi)).to_numpy(),
                              O2.scan(O2.OP_ADD_I32, xi))
        ctx.finalize()
        q.put((rank, "ok"))
    except BaseException:   # noqa: BLE001 - reported to the parent
        import traceback
        q.put((rank, traceback.format_exc()))


def test_ipc_ranks_on_two_gpus():
    if ngpus() < 2:
        pytest.skip("needs 2 GPUs")
    os.environ["SKL_COMM"] = "ipc"
    try:
        nid = S.Context.nccl_unique_id()
    finally:
        os.environ.pop("SKL_COMM", None)
    ctxm = mp.get_context("spawn")
    q = ctxm.Queue()
    procs = [ctxm.Process(target=_ipc_worker, args=(r, 2, nid, q)) for r in range(2)]
    for p in procs:
        p.start()
    res = {}
    try:
        for _ in range(2):
            r, msg = q.get(timeout=300)
            res[r] = msg
    finally:
        for p in procs:
            p.join(timeout=60)
            if p.is_alive():
                p.kill()
    assert res == {0: "ok", 1: "ok"}, res
