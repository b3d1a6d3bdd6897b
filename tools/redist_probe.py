import sys, time, numpy as np, torch
import os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from paper_conf_pact_steuwerg13_b200 import skl as S, apps as A, inputs as I
G, nvox = 4, 150**3
c4 = S.Context(G, devices=[0]*G)
st = torch.cuda.Stream(); torch.cuda.set_stream(st)
for g in range(G): c4.set_stream(g, st.cuda_stream)
img = I.uniform_f32(1, nvox)
w = S.Vector.from_numpy(c4, img).set_distribution(S.BLOCK)
v = S.Vector(c4, S.F32, nvox).set_distribution(S.BLOCK)
ident = S.Map(c4, A.IDENT_F32, S.F32, S.F32)
for xk in (1, 0):
    c4.set_option("xfer_kernel", xk)
    for _ in range(3):
        ident(w, out=v); v.set_distribution(S.COPY); v.set_distribution(S.BLOCK)
    torch.cuda.synchronize()
    # host time per call
    hs = []
    for _ in range(10):
        ident(w, out=v)
        t0 = time.perf_counter(); v.set_distribution(S.COPY); t1 = time.perf_counter()
        v.set_distribution(S.BLOCK); t2 = time.perf_counter()
        hs.append((t1 - t0, t2 - t1))
    torch.cuda.synchronize()
    # GPU time with the host far ahead
    torch.cuda._sleep(int(50e6))
    ev = []
    for _ in range(10):
        ident(w, out=v)
        a = torch.cuda.Event(enable_timing=True); b = torch.cuda.Event(enable_timing=True)
        a.record(); v.set_distribution(S.COPY); b.record(); v.set_distribution(S.BLOCK)
        ev.append((a, b))
    torch.cuda.synchronize()
    print(f"xfer_kernel={xk}: host set COPY {np.median([h[0] for h in hs])*1e6:.1f} us, set BLOCK {np.median([h[1] for h in hs])*1e6:.1f} us; "
          f"GPU (host ahead) {np.median([a.elapsed_time(b) for a, b in ev])*1e3:.1f} us", flush=True)

# copy(+) -> block: host and GPU time of the combine step
addf = S.Reduce(c4, A.ADD, S.F32)
cv = S.Vector(c4, S.F32, nvox)
idx = S.Vector.from_numpy(c4, np.arange(nvox, dtype=np.int32)).set_distribution(S.COPY)
touch = S.Map(c4, "void touch(int i, float* c) { c[i] = 1.0f; }", S.I32, S.VOID, extra=[S.F32 | S.PTR])
c4.set_option("xfer_kernel", 1)


def prep():
    cv.set_distribution(S.COPY, 0, addf)
    cv.fill(0.0)
    touch(idx, (cv, S.WRITE))


for _ in range(3):
    prep(); cv.set_distribution(S.BLOCK)
torch.cuda.synchronize()
hs = []
for _ in range(10):
    prep()
    t0 = time.perf_counter(); cv.set_distribution(S.BLOCK); hs.append(time.perf_counter() - t0)
torch.cuda.synchronize()
torch.cuda._sleep(int(50e6))
ev = []
for _ in range(10):
    prep()
    a = torch.cuda.Event(enable_timing=True); b = torch.cuda.Event(enable_timing=True)
    a.record(); cv.set_distribution(S.BLOCK); b.record()
    ev.append((a, b))
torch.cuda.synchronize()
print(f"copy(+)->block: host {np.median(hs)*1e6:.1f} us; GPU (host ahead) {np.median([a.elapsed_time(b) for a, b in ev])*1e3:.1f} us; "
      f"ok={bool(np.all(cv.to_numpy() == float(G)))}", flush=True)
