import sys
import numpy as np
sys.path.insert(0, "/root/repo"); sys.path.insert(0, "/root/repo/tests")
import test_gpu_fuzz as F
from paper_conf_pact_steuwerg13_b200 import skl as S, apps as A
# monkeypatch Reduce.__call__ to print state when called on a deferred Zip of (v, v)
orig_prog = F._program
G, seed = int(sys.argv[1]), int(sys.argv[2])
rng_steps = []
class Spy:
    pass
import oracle as O
real_assert = None
def run():
    rng = np.random.default_rng(seed)
    ctx = S.Context(G, devices=[0] * G)
    neg = S.Map(ctx, A.NEG, S.F32, S.F32); sq = S.Map(ctx, A.SQP1, S.F32, S.F32)
    add = S.Zip(ctx, A.ADD, S.F32, S.F32, S.F32); red = S.Reduce(ctx, A.SUM, S.F32)
    box = S.MapOverlap(ctx, A.BOX3, S.F32, S.F32, 1, S.NEAREST, 0.0)
    n = F.SIZES[rng.integers(len(F.SIZES))]
    vecs = [S.Vector(ctx, S.F32, n) for _ in range(3)]
    shadow = [np.zeros(n, np.float32) for _ in range(3)]
    for v in vecs: v.fill(0.0)
    mat = [S.Matrix(ctx, S.F32, F.ROWS, F.COLS) for _ in range(2)]
    mshadow = [np.zeros((F.ROWS, F.COLS), np.float32) for _ in range(2)]
    for m in mat: m.fill(0.0)
    dists = [(S.BLOCK, 0), (S.COPY, 0), (S.SINGLE, G - 1), (S.OVERLAP, 1), (S.BLOCK, 0)]
    for step in range(60):
        op = int(rng.integers(11)); i, j, k = (int(x) for x in rng.integers(3, size=3))
        desc = (op, i, j, k)
        if op == 0:
            x = (rng.random(n, dtype=np.float32) - np.float32(0.5)); vecs[i].copy_in(x); shadow[i] = x
        elif op == 1:
            d, a = dists[int(rng.integers(len(dists)))]; vecs[i].set_distribution(d, a); desc += ("dist", d, a)
        elif op == 2:
            f, ref = (neg, O.OM_NEG_F32) if rng.random() < 0.5 else (sq, O.OM_SQP1_F32)
            if i == j: F._no_overlap(vecs[i])
            f(vecs[i], out=vecs[j]); shadow[j] = O.map_(ref, shadow[i])
        elif op == 3:
            if k == i: F._no_overlap(vecs[i])
            add(vecs[i], vecs[j], out=vecs[k]); shadow[k] = O.zip_(O.OZ_ADD_F32, shadow[i], shadow[j])
        elif op == 4:
            got = neg(sq(vecs[i])).to_numpy()
        elif op == 5:
            st = [v.distribution() for v in vecs]
            got = float(red(add(vecs[i], vecs[j])).scalar())
            ref = O.reduce_(O.OP_ADD_F32, O.zip_(O.OZ_ADD_F32, shadow[i], shadow[j]))
            bad = abs(got - ref) > 1e-5 * max(1.0, float(np.abs(shadow[i]).sum() + np.abs(shadow[j]).sum()))
            print(step, desc, "dists", st, "got", got, "ref", ref, "BAD" if bad else "")
            if bad:
                print(" to_numpy sums", [float(v.to_numpy().astype(np.float64).sum()) for v in vecs])
                print(" shadow sums", [float(s.astype(np.float64).sum()) for s in shadow])
                t = S.Vector(ctx, S.F32, n); add(vecs[i], vecs[j], out=t)
                print(" unfused", float(red(t).scalar()), "red(vi)", float(red(vecs[i]).scalar()), "red(vj)", float(red(vecs[j]).scalar()))
                print(" again fused", float(red(add(vecs[i], vecs[j])).scalar()))
                return
        elif op == 6: pass
        elif op == 7:
            val = float(rng.integers(-3, 4)); vecs[i].fill(val); shadow[i] = np.full(n, val, np.float32); desc += ("fill", val)
        elif op == 8:
            a_, b_ = i % 2, 1 - i % 2; box(mat[a_], out=mat[b_]); mshadow[b_] = O.mapoverlap2d(O.OS_BOX3, mshadow[a_], 1, O.OB_NEAREST, 0.0)
        elif op == 9:
            if rng.random() < 0.5:
                x = rng.random((F.ROWS, F.COLS), dtype=np.float32); mat[i % 2].copy_in(x); mshadow[i % 2] = x
            else:
                F._no_overlap(mat[i % 2]); neg(mat[i % 2], out=mat[i % 2]); mshadow[i % 2] = -mshadow[i % 2]
        elif op == 10:
            if rng.random() < 0.5: pass
            else:
                d, a2 = dists[int(rng.integers(len(dists)))]; mat[i % 2].set_distribution(d, a2)
        if op in (0, 1, 7): print(step, desc, [v.distribution() for v in vecs])
run()
