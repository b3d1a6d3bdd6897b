"""Iterated Listing 1.5 Sobel probe on one GPU: microseconds per call for the three
ping-pong directions of an iterated 8192^2 stencil, and the output statistics."""
import sys, numpy as np, torch
import os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from paper_conf_pact_steuwerg13_b200 import skl as S, apps as A, inputs as I
ctx = S.Context(1)
st = torch.cuda.Stream(); torch.cuda.set_stream(st); ctx.set_stream(0, st.cuda_stream)
img = I.image_u8(5, 8192, 8192)
sob = S.MapOverlap(ctx, A.SOBEL, S.U8, S.U8, 1, S.NEUTRAL, 0)
a = S.Matrix.from_numpy(ctx, img); b = S.Matrix(ctx, S.U8, 8192, 8192); t = S.Matrix(ctx, S.U8, 8192, 8192)
sob(a, out=b); sob(b, out=t); sob(t, out=b)
torch.cuda.synchronize()
for name, fn in (("a->b", lambda: sob(a, out=b)), ("b->t", lambda: sob(b, out=t)), ("t->b", lambda: sob(t, out=b))):
    l0, p0 = ctx.counter("launches"), ctx.counter("p2p_bytes")
    torch.cuda._sleep(int(5e6))
    es = []
    for _ in range(10):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(); fn(); e1.record(); es.append((e0, e1))
    torch.cuda.synchronize()
    print(name, "launches/call", (ctx.counter("launches") - l0) / 10, "p2p", ctx.counter("p2p_bytes") - p0,
          "us", np.median([x.elapsed_time(y) for x, y in es]) * 1e3, flush=True)
# content statistics: fraction of zeros / 255 after 1 and 2 iterations
o1 = b.to_numpy()
print("iter-out zeros", float((o1 == 0).mean()), "sat", float((o1 == 255).mean()))
