"""LM OSEM Map launch configurations on one GPU: 10^7 events ordered longest
walk first (the bench's step), one Map into a zeroed copy(+) image, timed with
CUDA events (median of 5), checked against the oracle on a 1/50 sample.

  LM_CFGS="block,unroll,interleave,il_elems;..."
"""
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import oracle as O  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import apps as A  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import inputs as I  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import skl as S  # noqa: E402
from paper_conf_pact_steuwerg13_b200.lmosem import ListModeOSEM  # noqa: E402

N, NEV = 150, 10_000_000
events = I.lmosem_events(I.SEED_LMOSEM, NEV, N)
order = ListModeOSEM.path_order(events, N)
sorted_ev = np.ascontiguousarray(events[order])
sub = events[::50].copy()
c_ref = O.lmosem(sub, N, np.ones(N ** 3, np.float32))[0]
for cfg in os.environ.get("LM_CFGS", "256,1,0,0;128,1,0,0;128,1,1,1;256,1,1,1;64,1,1,1").split(";"):  # noqa: E501
    bt, un, il, j = (int(v) for v in cfg.split(","))
    ctx = S.Context(1)
    st = torch.cuda.Stream()
    torch.cuda.set_stream(st)
    ctx.set_stream(0, st.cuda_stream)
    for k, v in (("block_threads", bt), ("map_unroll", un), ("map_interleave", il), ("map_il_elems", j)):
        ctx.set_option(k, v)
    evd = ctx.struct_type("Event", A.EVENT_DECL, A.EVENT_SIZE, 4)
    lm = S.Map(ctx, A.lmosem_map(N), evd, S.VOID, extra=[S.F32 | S.PTR, S.F32 | S.PTR])
    addf = S.Reduce(ctx, A.ADD, S.F32)
    ev = S.Vector(ctx, evd, NEV).set_distribution(S.BLOCK)
    ev.copy_in(sorted_ev)
    f = S.Vector.from_numpy(ctx, np.ones(N ** 3, np.float32)).set_distribution(S.COPY)
    c = S.Vector(ctx, S.F32, N ** 3).set_distribution(S.COPY, 0, addf)
    ts = []
    for it in range(7):
        c.fill(0.0)
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        lm(ev, f, (c, S.WRITE))
        b.record()
        if it >= 2:
            ts.append((a, b))
    torch.cuda.synchronize()
    ms = float(np.median([x.elapsed_time(y) for x, y in ts]))
    evs = S.Vector(ctx, evd, sub.shape[0]).set_distribution(S.BLOCK)
    evs.copy_in(sub)
    c.fill(0.0)
    lm(evs, f, (c, S.WRITE))
    c.set_distribution(S.BLOCK)
    e = float(np.linalg.norm(c.to_numpy().astype(np.float64) - c_ref) / np.linalg.norm(c_ref))
    print(f"lmosem block={bt} unroll={un} interleave={il} il_elems={j}: {ms:.3f} ms  rel_l2={e:.2e}", flush=True)
    ctx.finalize()
