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
        # divergent per-event work: one event per thread (interleaved kernel with
        # one element per lane; 5.77 -> 5.67 ms for 10^7 events, tools/lmosem_probe.py)
        ctx.set_option("map_unroll", 1)
        ctx.set_option("map_interleave", 1)
        ctx.set_option("map_il_elems", 1)
        self.walk = S.Map(ctx, A.lmosem_map(N), self.evd, S.VOID, extra=[S.F32 | S.PTR, S.F32 | S.PTR])
        ctx.set_option("map_unroll", 4)
        ctx.set_option("map_interleave", 0)
        ctx.set_option("map_il_elems", 0)
        self.update = S.Zip(ctx, A.LMOSEM_UPDATE, S.F32, S.F32, S.F32)
        self.plus = S.Reduce(ctx, A.ADD, S.F32)
        n3 = N ** 3
        self.f = S.Vector(ctx, S.F32, n3).set_distribution(S.BLOCK)
        self.fn = S.Vector(ctx, S.F32, n3).set_distribution(S.BLOCK)
        self.c = S.Vector(ctx, S.F32, n3).set_distribution(S.COPY, 0, self.plus)
        self.subsets: list[S.Vector] = []

    @staticmethod
    def path_order(events: np.ndarray, N: int) -> np.ndarray:
        """A permutation of the events, longest ray walk first (application-level
        load balancing; within a subset the order of events does not change the
        result beyond fp32 atomic rounding).  The walk length is estimated on the
        host in float64 from the ray's entry and exit voxels (the number of voxel
        boundaries crossed + 1; 0 for rays that miss the volume).  Warps then hold
        rays of similar length, so fewer lanes idle while the longest ray of the
        warp finishes, and the block scheduler runs the long rays first."""
        ev = np.asarray(events, dtype=np.float64)
        p0, d = ev[:, 0:3], ev[:, 3:6] - ev[:, 0:3]
        amin = np.zeros(len(ev))
        amax = np.ones(len(ev))
        hit = np.ones(len(ev), dtype=bool)
        with np.errstate(divide="ignore", invalid="ignore"):
            for a in range(3):
                flat = d[:, a] == 0.0
                hit &= ~(flat & ((p0[:, a] < 0.0) | (p0[:, a] > N)))
                a0 = np.where(flat, -np.inf, (0.0 - p0[:, a]) / d[:, a])
                aN = np.where(flat, np.inf, (N - p0[:, a]) / d[:, a])
                amin = np.maximum(amin, np.minimum(a0, aN))
                amax = np.minimum(amax, np.maximum(a0, aN))
        hit &= amax > amin
        top = np.nextafter(float(N), 0.0)
        ent = np.clip(p0 + amin[:, None] * d, 0.0, top)
        ext = np.clip(p0 + amax[:, None] * d, 0.0, top)
        steps = np.abs(np.floor(ext) - np.floor(ent)).sum(axis=1) + 1.0
        key = np.where(hit, steps, 0.0)
        return np.argsort(-key, kind="stable")

    @staticmethod
    def subset_bounds(nev: int, nsub: int):
        """contiguous slices [lo, hi) of the event stream, sizes differing by <= 1"""
        return [(nev * i // nsub, nev * (i + 1) // nsub) for i in range(nsub)]

    def load_events(self, events: np.ndarray, nsub: int, balance: bool = True):
        """upload the list-mode events once, one block-distributed Vector per
        subset (each subset's events ordered longest walk first if `balance`)"""
        for v in self.subsets:
            v.destroy()
        self.subsets = []
        for lo, hi in self.subset_bounds(events.shape[0], nsub):
            sub = events[lo:hi]
            if balance:
                order = self.path_order(sub, self.N)
                G = self.ctx.ndev
                if G > 1:
                    # deal the sorted rays round-robin so that every device's
                    # block holds an equal share of long and short rays
                    order = np.concatenate([order[g::G] for g in range(G)])
                sub = sub[order]
            v = S.Vector(self.ctx, self.evd, hi - lo).set_distribution(S.BLOCK)
            v.copy_in(np.ascontiguousarray(sub))
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
