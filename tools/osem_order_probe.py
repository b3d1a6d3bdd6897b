"""LM OSEM walk over 10^6 events: device time per event order (and 10^7 for reference)."""
import sys
import numpy as np
import torch
sys.path.insert(0, __file__.rsplit("/tools/", 1)[0])
from paper_conf_pact_steuwerg13_b200 import skl as S, inputs as I, apps as A
from paper_conf_pact_steuwerg13_b200.lmosem import ListModeOSEM

N = 150
ctx = S.Context(1)
st = torch.cuda.Stream(); torch.cuda.set_stream(st); ctx.set_stream(0, st.cuda_stream)
ctx.set_option("xfer_chunks", 1)
osem = ListModeOSEM(ctx, N)
osem.set_image(np.ones(N ** 3, np.float32))
osem.f.set_distribution(S.COPY)
osem.c.set_distribution(S.COPY, 0, osem.plus)


def t_walk(evs, reps=5):
    v = S.Vector(ctx, osem.evd, evs.shape[0]).set_distribution(S.BLOCK)
    v.copy_in(np.ascontiguousarray(evs))
    osem.walk(v, osem.f, (osem.c, S.WRITE))
    torch.cuda.synchronize()
    torch.cuda._sleep(int(20e6))
    es = []
    for _ in range(reps):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(); osem.walk(v, osem.f, (osem.c, S.WRITE)); b.record(); es.append((a, b))
    torch.cuda.synchronize()
    v.destroy()
    return float(np.median([a.elapsed_time(b) for a, b in es]))


ev = I.lmosem_events(I.SEED_LMOSEM, 10_000_000, N)
sub = ev[:1_000_000]
order = ListModeOSEM.path_order(sub, N)
print(f"10^6 generation order: {t_walk(sub):.3f} ms", flush=True)
print(f"10^6 longest first:   {t_walk(sub[order]):.3f} ms", flush=True)
print(f"10^6 shortest first:  {t_walk(sub[order[::-1]]):.3f} ms", flush=True)
hit = order[: int((ListModeOSEM.path_order(sub, N) is not None) and 0)]  # placeholder
for ways in (2, 4, 8):
    o2 = np.concatenate([order[g::ways] for g in range(ways)])
    print(f"10^6 longest first dealt {ways} ways: {t_walk(sub[o2]):.3f} ms", flush=True)
full_order = ListModeOSEM.path_order(ev, N)
t10 = t_walk(ev[full_order], reps=3)
print(f"10^7 longest first:   {t10:.3f} ms  ({t10 / 10:.3f} ms per 10^6)", flush=True)
for bt in (128, 512):
    ctx.set_option("block_threads", bt)
    ctx.set_option("map_unroll", 1)
    osem.walk = S.Map(ctx, A.lmosem_map(N), osem.evd, S.VOID, extra=[S.F32 | S.PTR, S.F32 | S.PTR])
    print(f"block {bt}: 10^6 longest first {t_walk(sub[order]):.3f} ms", flush=True)
