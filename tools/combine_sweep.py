"""copy(+) -> block of a 150^3 fp32 Vector on G logical devices of one GPU:
device time of the fold per (combine_peer, combine_unroll, block_threads).
COMB_CFGS="peer,unroll,block;..." """
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from paper_conf_pact_steuwerg13_b200 import apps as A  # noqa: E402
from paper_conf_pact_steuwerg13_b200 import skl as S  # noqa: E402

G, nvox = int(os.environ.get("COMB_G", "4")), 150 ** 3
flush = torch.empty(64 << 20, dtype=torch.float32, device="cuda")
clean = torch.zeros(64 << 20, dtype=torch.float32, device="cuda")
sink = torch.zeros((), dtype=torch.float32, device="cuda")
for cfg in os.environ.get("COMB_CFGS", "1,2,256").split(";"):
    peer, unr, bt = (int(x) for x in cfg.split(","))
    c = S.Context(G, devices=[0] * G)
    st = torch.cuda.Stream()
    torch.cuda.set_stream(st)
    for g in range(G):
        c.set_stream(g, st.cuda_stream)
    c.set_option("combine_peer", peer)
    c.set_option("combine_unroll", unr)
    c.set_option("block_threads", bt)
    addf = S.Reduce(c, A.ADD, S.F32)
    cv = S.Vector(c, S.F32, nvox)
    idx = S.Vector.from_numpy(c, np.arange(nvox, dtype=np.int32)).set_distribution(S.BLOCK)
    touch = S.Map(c, "void touch(int i, float* c) { c[i] = 1.0f; }", S.I32, S.VOID, extra=[S.F32 | S.PTR])
    ts = []
    for it in range(13):
        cv.set_distribution(S.COPY, 0, addf)
        cv.fill(0.0)
        touch(idx, (cv, S.WRITE))
        flush.zero_()               # evict, then read a clean buffer: the fold starts
        sink.copy_(clean.sum())     # cold and without dirty lines to write back (as bench.py)
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        cv.set_distribution(S.BLOCK)
        b.record()
        if it >= 3:
            ts.append((a, b))
    torch.cuda.synchronize()
    ok = bool(np.all(cv.to_numpy() == 1.0))
    ms = float(np.median([a.elapsed_time(b) for a, b in ts]))
    print(f"combine G={G} peer={peer} unroll={unr} block={bt}: {ms * 1e3:.1f} us  "
          f"{(G + 1) * nvox * 4 / (ms / 1e3) / 1e9:.0f} GB/s (fold traffic, cold)  ok={ok}", flush=True)
    c.finalize()
