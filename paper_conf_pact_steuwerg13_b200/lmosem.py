"""List-mode OSEM reconstruction over several subsets (
reading A29), written as a SkelCL user program: every step is a skeleton call
or a redistribution of the library, nothing is computed here.

Per subset l (events E_l, a contiguous slice of the list-mode stream):
  1. f: block -> copy (all-gather over the devices); c: copy(+), zeroed
  2. Map over E_l (block): fp = sum_k len_k f[v_k]; if fp > 0, c[v_k] += len_k / fp
  3. c: copy(+) -> block (the replicas are summed, A25); f: copy -> block (no move)
  4. f <- f * c (Zip, block; sensitivity 1, A29)
so f changes distribution twice and c once every subset: the redistribution
machinery runs at every iteration, as in the paper's application.
"""
from __future__ import annotations

import numpy as np

from . import apps as A
from . import skl as S


class ListModeOSEM:
    def __init__(self, ctx: S.Context, N: int):
        self.ctx, self.N = ctx, N
        self.evd = ctx.struct_type("Event", A.EVENT_DECL, A.EVENT_SIZE, 4)
        ctx.set_option("map_unroll", 1)   # divergent per-event work: one chunk per thread
        self.walk = S.Map(ctx, A.lmosem_map(N), self.evd, S.VOID, extra=[S.F32 | S.PTR, S.F32 | S.PTR])
        ctx.set_option("map_unroll", 4)
        self.update = S.Zip(ctx, A.LMOSEM_UPDATE, S.F32, S.F32, S.F32)
        self.plus = S.Reduce(ctx, A.ADD, S.F32)
        n3 = N ** 3
        self.f = S.Vector(ctx, S.F32, n3).set_distribution(S.BLOCK)
        self.fn = S.Vector(ctx, S.F32, n3).set_distribution(S.BLOCK)
        self.c = S.Vector(ctx, S.F32, n3).set_distribution(S.COPY, 0, self.plus)
        self.subsets: list[S.Vector] = []

    @staticmethod
    def subset_bounds(nev: int, nsub: int):
        """contiguous slices [lo, hi) of the event stream, sizes differing by <= 1"""
        return [(nev * i // nsub, nev * (i + 1) // nsub) for i in range(nsub)]

    def load_events(self, events: np.ndarray, nsub: int):
        """upload the list-mode events once, one block-distributed Vector per subset"""
        for v in self.subsets:
            v.destroy()
        self.subsets = []
        for lo, hi in self.subset_bounds(events.shape[0], nsub):
            v = S.Vector(self.ctx, self.evd, hi - lo).set_distribution(S.BLOCK)
            v.copy_in(np.ascontiguousarray(events[lo:hi]))
            self.subsets.append(v)

    def set_image(self, f0: np.ndarray):
        self.f.copy_in(np.ascontiguousarray(f0, dtype=np.float32))

    def subset_step(self, ev: S.Vector):
        f, c = self.f, self.c
        f.set_distribution(S.COPY)                 # 1. all-gather the image
        c.set_distribution(S.COPY, 0, self.plus)
        c.fill(0.0)
        self.walk(ev, f, (c, S.WRITE))             # 2. Map over the subset's events
        c.set_distribution(S.BLOCK)                # 3. copy(+) -> block combine
        f.set_distribution(S.BLOCK)
        self.update(f, c, out=self.fn)             # 4. f <- f * c
        self.f, self.fn = self.fn, self.f

    def iterate(self, passes: int = 1):
        """`passes` full passes over all subsets"""
        for _ in range(passes):
            for ev in self.subsets:
                self.subset_step(ev)

    def image(self) -> np.ndarray:
        return self.f.to_numpy()

    def destroy(self):
        for v in self.subsets + [self.f, self.fn, self.c]:
            v.destroy()
        self.subsets = []
