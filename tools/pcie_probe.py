"""PCIe floor of the end-to-end Mandelbrot step on one GPU: pinned host <->
device copies of the step's bytes (96 MiB in, 48 MiB out), each direction alone
and both at once on two streams (full duplex), median of 10."""
import numpy as np
import torch

MB = 1 << 20
hin = torch.empty(96 * MB, dtype=torch.uint8).pin_memory()
hout = torch.empty(48 * MB, dtype=torch.uint8).pin_memory()
din = torch.empty(96 * MB, dtype=torch.uint8, device="cuda")
dout = torch.empty(48 * MB, dtype=torch.uint8, device="cuda")
s1, s2 = torch.cuda.Stream(), torch.cuda.Stream()


def run(fn, reps=10):
    ts = []
    for _ in range(reps + 2):
        torch.cuda.synchronize()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        s1.wait_event(a)
        s2.wait_event(a)
        fn()
        e1, e2 = torch.cuda.Event(), torch.cuda.Event()
        e1.record(s1)
        e2.record(s2)
        torch.cuda.current_stream().wait_event(e1)
        torch.cuda.current_stream().wait_event(e2)
        b.record()
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b))
    return float(np.median(ts[2:]))


def h2d():
    with torch.cuda.stream(s1):
        din.copy_(hin, non_blocking=True)


def d2h():
    with torch.cuda.stream(s2):
        hout.copy_(dout, non_blocking=True)


def both():
    h2d()
    d2h()


for name, fn in (("H2D 96 MiB", h2d), ("D2H 48 MiB", d2h), ("both at once", both)):
    print(f"{name:14s} {run(fn):.3f} ms", flush=True)
