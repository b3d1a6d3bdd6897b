"""The one-process-per-GPU mode (skl_init_dist) with 2 and 3 ranks, run as
processes on one GPU, over the shared-memory loopback transport (SKL_COMM=shm;
NCCL refuses two ranks on one device) and over the NVLink peer-memory transport
(SKL_COMM=ipc: IPC heap, in-kernel peer loads/stores, device barriers - on one
GPU the "peers" are the other processes' allocations of the same device).  Everything above the transport is the
multi-rank code path: rank-local parts, the canonical transfer lists executed
by both ranks, cross-rank Reduce / Scan carry-in, halo exchange, copy(+) ->
block combine, collective host reads.  Each rank checks the oracle."""
import multiprocessing as mp
import os
import sys
import traceback

import numpy as np
import pytest

from gpu_util import require_gpu

pytestmark = pytest.mark.gpu

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _worker(rank, world, nid, q, comm="shm"):
    try:
        os.environ["SKL_COMM"] = comm
        sys.path.insert(0, ROOT)
        sys.path.insert(0, os.path.join(ROOT, "tests"))
        import oracle as O
        from paper_conf_pact_steuwerg13_b200 import apps as A
        from paper_conf_pact_steuwerg13_b200 import inputs as I
        from paper_conf_pact_steuwerg13_b200 import skl as S
        from paper_conf_pact_steuwerg13_b200.lmosem import ListModeOSEM
        if comm == "nccl":   # as in the bench: torch (with its own NCCL) in the same process
            import torch
            torch.zeros(1, device="cuda")

        def rel(a, b):
            a, b = np.asarray(a, np.float64), np.asarray(b, np.float64)
            return float(np.linalg.norm(a - b) / max(np.linalg.norm(b), 1e-300))

        ctx = S.Context.dist(rank, world, 0, nid)
        assert ctx.devices() == (world, rank, 1)
        n = 100003
        x = I.uniform_f32(1, n)
        y = I.uniform_f32(2, n)
        vx, vy = S.Vector.from_numpy(ctx, x), S.Vector.from_numpy(ctx, y)
        # Zip + Reduce across ranks (ordered combine of the two partials)
        d = float(S.Reduce(ctx, A.SUM, S.F32)(S.Zip(ctx, A.MULT, S.F32, S.F32, S.F32)(vx, vy)).scalar())
        ref = O.reduce_(O.OP_ADD_F32, O.zip_(O.OZ_MULT_F32, x, y))
        assert abs(d - ref) <= 1e-5 * abs(ref), (d, ref)
        r = S.Reduce(ctx, A.RIGHT_F32, S.F32)(vx).scalar()     # order across ranks
        assert r == x[-1]
        assert S.Reduce(ctx, A.LEFT_F32, S.F32)(vx).scalar() == x[0]
        # Scan with carry-in from rank 0 to rank 1
        xi = I.uniform_int(3, n, -1000, 1000)
        assert np.array_equal(S.Scan(ctx, A.ADD_I32, S.I32)(S.Vector.from_numpy(ctx, xi)).to_numpy(),
                              O.scan(O.OP_ADD_I32, xi))
        # Map (collective download)
        assert np.array_equal(S.Map(ctx, A.SQP1, S.F32, S.F32)(vx).to_numpy(), O.map_(O.OM_SQP1_F32, x))
        # distributions: block -> copy -> single(1) -> overlap -> block
        v = S.Vector.from_numpy(ctx, x)
        for dd, arg in ((S.BLOCK, 0), (S.COPY, 0), (S.SINGLE, world - 1), (S.OVERLAP, 5), (S.BLOCK, 0)):
            v.set_distribution(dd, arg)
            assert np.array_equal(v.to_numpy(), x), (dd, arg)
        # MapOverlap with a halo exchange between the ranks, twice (halo refresh)
        img = I.image_f32(I.SEED_GAUSS, 97, 61)
        gau = S.MapOverlap(ctx, A.gaussian5(), S.F32, S.F32, 2, S.NEAREST, 0.0)
        h0 = ctx.counter("halo_push_bytes")
        g2 = gau(gau(S.Matrix.from_numpy(ctx, img)))
        r1 = O.mapoverlap2d(O.OS_GAUSS5, img, 2, O.OB_NEAREST, 0.0)
        assert np.array_equal(g2.to_numpy(), O.mapoverlap2d(O.OS_GAUSS5, r1, 2, O.OB_NEAREST, 0.0))
        if comm == "ipc" and world > 1:   # the first stencil pushed its border rows into the neighbours' halos
            assert ctx.counter("halo_push_bytes") > h0
        # iterated Sobel (ping-pong, halos pushed / exchanged every iteration)
        im8 = I.image_u8(I.SEED_SOBEL, 131, 80)
        sob = S.MapOverlap(ctx, A.SOBEL_TUNED, S.U8, S.U8, 1, S.NEUTRAL, 0)
        a8 = S.Matrix.from_numpy(ctx, im8)
        b8, t8 = sob(a8), None
        ref8 = O.mapoverlap2d(O.OS_SOBEL, im8, 1, O.OB_NEUTRAL, 0)
        for _ in range(3):
            t8 = sob(b8, out=t8)
            b8, t8 = t8, b8
            ref8 = O.mapoverlap2d(O.OS_SOBEL, ref8, 1, O.OB_NEUTRAL, 0)
        assert np.array_equal(b8.to_numpy(), ref8)
        # copy(+) -> block: each rank adds its own events into its replica (LM OSEM)
        N, nev = 10, 3000
        osem = ListModeOSEM(ctx, N)
        ev = I.lmosem_events(I.SEED_LMOSEM, nev, N)
        f0 = np.ones(N ** 3, np.float32)
        osem.load_events(ev, 2)
        osem.set_image(f0)
        osem.iterate(1)
        f = f0
        for lo, hi in ListModeOSEM.subset_bounds(nev, 2):
            f = O.lmosem(ev[lo:hi], N, f)[1].astype(np.float32)
        assert rel(osem.image(), f) <= 1e-4
        osem.destroy()
        # Allpairs: A block over the ranks, B copied to both
        a = I.uniform_f32(8, 70 * 20).reshape(70, 20)
        b = I.uniform_f32(9, 30 * 20).reshape(30, 20)
        ap = S.Allpairs(ctx, A.MULT, S.F32, S.F32, reduce=A.ADD)
        assert np.array_equal(ap(S.Matrix.from_numpy(ctx, a), S.Matrix.from_numpy(ctx, b)).to_numpy(),
                              O.allpairs(O.AP_DOT, a, b))
        if comm == "nccl":   # the NCCL transport is the one set up
            assert ctx.counter("nccl_comm") == 1
            if world == 1:     # no move leaves the rank: no send/recv group is issued
                assert ctx.counter("nccl_groups") == 0
        ctx.finalize()
        q.put((rank, "ok"))
    except BaseException:   # noqa: BLE001 - reported to the parent
        q.put((rank, traceback.format_exc()))


@pytest.mark.parametrize("world", [2, 3])
@pytest.mark.parametrize("comm", ["shm", "ipc"])
def test_ranks_on_one_gpu(world, comm):
    require_gpu()
    sys.path.insert(0, ROOT)
    from paper_conf_pact_steuwerg13_b200 import skl as S
    os.environ["SKL_COMM"] = comm
    try:
        nid = S.Context.nccl_unique_id()
    finally:
        os.environ.pop("SKL_COMM", None)
    assert nid.startswith(b"/skl_")
    ctxm = mp.get_context("spawn")
    q = ctxm.Queue()
    procs = [ctxm.Process(target=_worker, args=(r, world, nid, q, comm)) for r in range(world)]
    for p in procs:
        p.start()
    results = {}
    try:
        for _ in range(world):
            rank, msg = q.get(timeout=600)
            results[rank] = msg
    finally:
        for p in procs:
            p.join(timeout=60)
            if p.is_alive():
                p.kill()
    assert results == {r: "ok" for r in range(world)}, results


@pytest.mark.parametrize("comm", ["nccl", "ipc", "shm"])
def test_one_rank_forced_dist(comm):
    """world size 1 with SKL_DIST_FORCE=1: the multi-process code path and its
    transport on one GPU - for NCCL (which refuses two ranks on one device) the
    library's libnccl load, ncclGetUniqueId, ncclCommInitRank and ncclCommDestroy
    next to torch (and torch's NCCL) in the same process - with every oracle
    check of the multi-rank worker"""
    require_gpu()
    sys.path.insert(0, ROOT)
    from paper_conf_pact_steuwerg13_b200 import skl as S
    os.environ["SKL_COMM"] = comm
    os.environ["SKL_DIST_FORCE"] = "1"
    try:
        nid = S.Context.nccl_unique_id()
        ctxm = mp.get_context("spawn")
        q = ctxm.Queue()
        p = ctxm.Process(target=_worker, args=(0, 1, nid, q, comm))
        p.start()
        try:
            rank, msg = q.get(timeout=600)
        finally:
            p.join(timeout=60)
            if p.is_alive():
                p.kill()
    finally:
        os.environ.pop("SKL_COMM", None)
        os.environ.pop("SKL_DIST_FORCE", None)
    assert (rank, msg) == (0, "ok"), msg
