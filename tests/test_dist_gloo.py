"""Multi-process (world size 2, gloo, CPU) tests of the N>1 host logic.

In one-process-per-GPU mode every rank walks the same canonical transfer list
(skl_plan_transfers) inside one NCCL group and posts the send/recv halves that
touch it.  Here two CPU processes do exactly that with torch.distributed (gloo)
isend/irecv on host arrays standing in for the device parts, and check that
every rank ends with precisely its target layout (values = global indices, so a
misplaced unit is caught), and that the copy(+) -> block gather + GPU-order fold
(A25) equals the oracle's combine.  No GPU is involved.
"""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

from paper_conf_pact_steuwerg13_b200 import skl as S

DISTS = [(S.SINGLE, 0), (S.SINGLE, 1), (S.COPY, 0), (S.BLOCK, 0), (S.OVERLAP, 1), (S.OVERLAP, 4)]


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _layout(units, G, kind, arg, g, cols):
    lo, hi = S.plan_range(units, G, kind, arg, g, kind == S.OVERLAP)
    a = np.full((max(hi - lo, 0), cols), -1.0, np.float32)
    return lo, hi, a


def _redistribute(rank, G, units, cols, fk, fa, tk, ta):
    """one rank's side of a planned redistribution; returns (lo, hi, part)"""
    flo, fhi, src = _layout(units, G, fk, fa, rank, cols)
    # source part holds the right values (row u = u)
    src[:] = np.arange(flo, fhi, dtype=np.float32)[:, None]
    tlo, thi, dst = _layout(units, G, tk, ta, rank, cols)
    # units already present stay (local copy)
    a, b = max(flo, tlo), min(fhi, thi)
    if b > a:
        dst[a - tlo:b - tlo] = src[a - flo:b - flo]
    ops, bufs = [], []
    for s, su, d, du, n in S.plan_transfers(units, G, fk, fa, tk, ta):
        if s == rank and d != rank:
            t = torch.from_numpy(np.ascontiguousarray(src[su - flo:su - flo + n]))
            ops.append(dist.P2POp(dist.isend, t, d))
            bufs.append(t)
        elif d == rank and s != rank:
            t = torch.empty((n, cols), dtype=torch.float32)
            ops.append(dist.P2POp(dist.irecv, t, s))
            bufs.append((t, du))
    if ops:
        for r in dist.batch_isend_irecv(ops):
            r.wait()
    for x in bufs:
        if isinstance(x, tuple):
            t, du = x
            dst[du - tlo:du - tlo + t.shape[0]] = t.numpy()
    return tlo, thi, dst


def _worker(rank, G, port, q):
    try:
        os.environ["MASTER_ADDR"] = "127.0.0.1"
        os.environ["MASTER_PORT"] = str(port)
        dist.init_process_group("gloo", rank=rank, world_size=G)
        import oracle as O
        errors = []
        for units, cols in ((1, 1), (9, 3), (64, 2), (1001, 1)):
            for fk, fa in DISTS:
                for tk, ta in DISTS:
                    if (fk == S.SINGLE and fa >= G) or (tk == S.SINGLE and ta >= G):
                        continue
                    tlo, thi, dst = _redistribute(rank, G, units, cols, fk, fa, tk, ta)
                    want = np.repeat(np.arange(tlo, thi, dtype=np.float32)[:, None], cols, 1)
                    if not np.array_equal(dst, want):
                        errors.append((units, fk, fa, tk, ta, rank))
        # copy(+) -> block: all-to-all gather of replica slices, fold in GPU order
        n = 1000
        rep = (np.arange(n, dtype=np.int32) * (rank + 1)) % 97 - 48      # this rank's replica
        lo, hi = O.block_range(n, G, rank)
        stage = np.zeros((G, hi - lo), np.int32)
        ops, keep = [], []
        for g in range(G):                       # canonical order: dst-major, then src
            glo, ghi = O.block_range(n, G, g)
            for h in range(G):
                if h == rank and g != rank:
                    t = torch.from_numpy(rep[glo:ghi].copy())
                    ops.append(dist.P2POp(dist.isend, t, g))
                    keep.append(t)
                elif g == rank and h != rank:
                    t = torch.empty(ghi - glo, dtype=torch.int32)
                    ops.append(dist.P2POp(dist.irecv, t, h))
                    keep.append((t, h))
                elif g == rank and h == rank:
                    stage[h] = rep[glo:ghi]
        for r in dist.batch_isend_irecv(ops):
            r.wait()
        for x in keep:
            if isinstance(x, tuple):
                stage[x[1]] = x[0].numpy()
        all_reps = np.stack([(np.arange(n, dtype=np.int32) * (g + 1)) % 97 - 48 for g in range(G)])
        want = O.combine(O.OP_ADD_I32, all_reps)[lo:hi]
        got = O.combine(O.OP_ADD_I32, stage)
        if not np.array_equal(got, want):
            errors.append(("combine", rank))
        dist.barrier()
        dist.destroy_process_group()
        q.put((rank, errors))
    except Exception as e:  # pragma: no cover
        q.put((rank, [repr(e)]))


@pytest.mark.parametrize("G", [2])
def test_planned_transfers_over_gloo(G):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, G, port, q)) for r in range(G)]
    for p in procs:
        p.start()
    res = dict(q.get(timeout=300) for _ in range(G))
    for p in procs:
        p.join(timeout=60)
    for r in range(G):
        assert res[r] == [], res[r]
