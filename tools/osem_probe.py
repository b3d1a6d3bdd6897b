"""Per-step device times of one LM OSEM subset (10^6 events) vs the 10^7-event Map."""
import sys
import numpy as np
import torch
sys.path.insert(0, __file__.rsplit("/tools/", 1)[0])
from paper_conf_pact_steuwerg13_b200 import skl as S, inputs as I
from paper_conf_pact_steuwerg13_b200.lmosem import ListModeOSEM

N, nev, nsub = 150, 10_000_000, 10
ctx = S.Context(1)
st = torch.cuda.Stream(); torch.cuda.set_stream(st); ctx.set_stream(0, st.cuda_stream)
events = I.lmosem_events(I.SEED_LMOSEM, nev, N)
osem = ListModeOSEM(ctx, N)
osem.load_events(events, nsub)
osem.set_image(np.ones(N ** 3, np.float32))
f, c = osem.f, osem.c
for _ in range(2):
    osem.iterate(1)
torch.cuda.synchronize()
torch.cuda._sleep(int(100e6))
rows = []
for ev in osem.subsets:
    e = [torch.cuda.Event(enable_timing=True) for _ in range(6)]
    e[0].record()
    osem.f.set_distribution(S.COPY); osem.c.set_distribution(S.COPY, 0, osem.plus)
    osem.c.fill(0.0)
    e[1].record()
    osem.walk(ev, osem.f, (osem.c, S.WRITE))
    e[2].record()
    osem.c.set_distribution(S.BLOCK); osem.f.set_distribution(S.BLOCK)
    e[3].record()
    osem.update(osem.f, osem.c, out=osem.fn)
    e[4].record()
    osem.f, osem.fn = osem.fn, osem.f
    e[5].record()
    rows.append(e)
torch.cuda.synchronize()
t = np.array([[r[i].elapsed_time(r[i + 1]) * 1e3 for i in range(5)] for r in rows])
print("per subset us: fill/redist %.1f  map %.1f  combine %.1f  zip %.1f  swap %.1f" % tuple(t.mean(axis=0)))
print("map per subset:", np.round(t[:, 1], 1))
