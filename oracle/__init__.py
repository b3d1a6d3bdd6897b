"""ctypes front-end of the CPU oracle (oracle.cpp).

TEST INFRASTRUCTURE ONLY: only tests/, __graft_entry__.smoke() and bench.py's
cpu_baseline / --impl reference legs may import this package.  The product path
(paper_conf_pact_steuwerg13_b200) must never import it.

The arithmetic lives in oracle.cpp (plain single-threaded C++, -O2
-ffp-contract=off -fno-fast-math); this file only marshals numpy arrays.
"""
from __future__ import annotations

import ctypes as C
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "liboracle.so")
_SRC = os.path.join(_HERE, "oracle.cpp")

# enums mirrored from oracle.h
OM_NEG_F32, OM_SQP1_F32, OM_INV_U8, OM_AFFINE_I32 = range(4)
OZ_ADD_F32, OZ_MULT_F32, OZ_SUB_I32 = range(3)
OP_ADD_F32, OP_ADD_I32, OP_MAX_F32, OP_LEFT_F32, OP_RIGHT_F32, OP_AFFINE_U32 = range(6)
OS_IDENT, OS_SHIFT_X, OS_SHIFT_Y, OS_BOX3, OS_SOBEL, OS_GAUSS5 = range(6)
OB_NEUTRAL, OB_NEAREST = 0, 1

CFLAGS = ["-O2", "-ffp-contract=off", "-fno-fast-math", "-std=c++17", "-fPIC", "-shared"]


def build(force: bool = False) -> str:
    """Compile liboracle.so (also called by __graft_entry__.build())."""
    if force or not os.path.exists(_SO) or os.path.getmtime(_SO) < max(
            os.path.getmtime(_SRC), os.path.getmtime(os.path.join(_HERE, "oracle.h"))):
        subprocess.check_call(["g++", *CFLAGS, "-o", _SO, _SRC])
    return _SO


_lib = None


def lib():
    global _lib
    if _lib is None:
        build()
        L = C.CDLL(_SO)
        vp, sz = C.c_void_p, C.c_size_t
        L.oracle_map.argtypes = [C.c_int, vp, vp, sz]
        L.oracle_mandelbrot.argtypes = [vp, vp, sz, C.c_uint32]
        L.oracle_mandelbrot.restype = C.c_uint64
        L.oracle_row_sums.argtypes = [vp, sz, sz, vp]
        L.oracle_zip.argtypes = [C.c_int, vp, vp, vp, sz]
        L.oracle_reduce.argtypes = [C.c_int, vp, sz, vp]
        L.oracle_scan.argtypes = [C.c_int, vp, sz, vp]
        L.oracle_combine.argtypes = [C.c_int, vp, C.c_int, sz, vp]
        L.oracle_mapoverlap2d.argtypes = [C.c_int, C.c_int, vp, vp, sz, sz, C.c_int, C.c_int, vp]
        L.oracle_mapoverlap1d.argtypes = [C.c_int, vp, vp, sz, C.c_int, C.c_int, C.c_float]
        L.oracle_gauss5_weights.argtypes = [vp]
        L.oracle_block_range.argtypes = [sz, C.c_int, C.c_int, C.POINTER(sz), C.POINTER(sz)]
        L.oracle_overlap_range.argtypes = [sz, C.c_int, C.c_int, sz, C.POINTER(sz), C.POINTER(sz)]
        L.oracle_siddon.argtypes = [vp, vp, C.c_int, vp, vp, sz]
        L.oracle_siddon.restype = sz
        L.oracle_lmosem.argtypes = [vp, sz, C.c_int, vp, vp, vp, C.POINTER(C.c_uint64)]
        L.oracle_lmosem.restype = C.c_uint64
        for f in ("oracle_map", "oracle_zip", "oracle_reduce", "oracle_scan", "oracle_combine",
                  "oracle_mapoverlap2d", "oracle_mapoverlap1d"):
            getattr(L, f).restype = C.c_int
        _lib = L
    return _lib


def _p(a: np.ndarray):
    assert a.flags["C_CONTIGUOUS"]
    return a.ctypes.data_as(C.c_void_p)


_MAP_T = {OM_NEG_F32: (np.float32, np.float32), OM_SQP1_F32: (np.float32, np.float32),
          OM_INV_U8: (np.uint8, np.uint8), OM_AFFINE_I32: (np.int32, np.int32)}


def map_(fn: int, x: np.ndarray) -> np.ndarray:
    ti, to = _MAP_T[fn]
    x = np.ascontiguousarray(x, dtype=ti)
    y = np.empty(x.shape, dtype=to)
    assert lib().oracle_map(fn, _p(x), _p(y), x.size) == 0
    return y


def mandelbrot(c: np.ndarray, max_iter: int):
    """c: float32 [..., 2]; returns (uint32 counts [...], total iterations)."""
    c = np.ascontiguousarray(c, dtype=np.float32)
    out = np.empty(c.shape[:-1], dtype=np.uint32)
    tot = lib().oracle_mandelbrot(_p(c), _p(out), out.size, max_iter)
    return out, int(tot)


def row_sums(counts: np.ndarray) -> np.ndarray:
    counts = np.ascontiguousarray(counts, dtype=np.uint32)
    s = np.empty(counts.shape[0], dtype=np.uint64)
    lib().oracle_row_sums(_p(counts), counts.shape[0], counts.shape[1], _p(s))
    return s


_ZIP_T = {OZ_ADD_F32: np.float32, OZ_MULT_F32: np.float32, OZ_SUB_I32: np.int32}


def zip_(fn: int, l: np.ndarray, r: np.ndarray) -> np.ndarray:
    t = _ZIP_T[fn]
    l = np.ascontiguousarray(l, dtype=t)
    r = np.ascontiguousarray(r, dtype=t)
    if l.size != r.size:
        raise ValueError("zip: size mismatch")
    y = np.empty(l.shape, dtype=t)
    assert lib().oracle_zip(fn, _p(l), _p(r), _p(y), l.size) == 0
    return y


# element dtype in, result dtype out; affine pairs are uint32 [..., 2]
_OP_T = {OP_ADD_F32: (np.float32, np.float64), OP_ADD_I32: (np.int32, np.int32),
         OP_MAX_F32: (np.float32, np.float32), OP_LEFT_F32: (np.float32, np.float32),
         OP_RIGHT_F32: (np.float32, np.float32), OP_AFFINE_U32: (np.uint32, np.uint32)}


def _nelem(op, x):
    return x.shape[0]


def reduce_(op: int, x: np.ndarray):
    ti, to = _OP_T[op]
    x = np.ascontiguousarray(x, dtype=ti)
    n = _nelem(op, x)
    out = np.empty((2,) if op == OP_AFFINE_U32 else (1,), dtype=to)
    rc = lib().oracle_reduce(op, _p(x), n, _p(out))
    if rc == -1:
        raise ValueError("reduce of an empty vector (A11)")
    assert rc == 0
    return out if op == OP_AFFINE_U32 else out[0]


def scan(op: int, x: np.ndarray) -> np.ndarray:
    ti, to = _OP_T[op]
    x = np.ascontiguousarray(x, dtype=ti)
    n = _nelem(op, x)
    out = np.empty(x.shape, dtype=to)
    rc = lib().oracle_scan(op, _p(x), n, _p(out))
    if rc == -1:
        raise ValueError("scan of an empty vector")
    assert rc == 0
    return out


def combine(op: int, replicas: np.ndarray) -> np.ndarray:
    """replicas: [G, n] (or [G, n, 2] for affine) -> [n] folded in GPU order."""
    ti, to = _OP_T[op]
    replicas = np.ascontiguousarray(replicas, dtype=ti)
    G, n = replicas.shape[0], replicas.shape[1]
    out = np.empty(replicas.shape[1:], dtype=to)
    assert lib().oracle_combine(op, _p(replicas), G, n, _p(out)) == 0
    return out


def mapoverlap2d(stencil: int, img: np.ndarray, d: int, boundary: int, neutral=0):
    if img.dtype == np.uint8:
        t, nv = 0, np.array([neutral], dtype=np.uint8)
    else:
        img = img.astype(np.float32, copy=False)
        t, nv = 1, np.array([neutral], dtype=np.float32)
    img = np.ascontiguousarray(img)
    out = np.empty_like(img)
    assert lib().oracle_mapoverlap2d(stencil, t, _p(img), _p(out), img.shape[0], img.shape[1],
                                     d, boundary, _p(nv)) == 0
    return out


def mapoverlap1d(stencil: int, v: np.ndarray, d: int, boundary: int, neutral: float = 0.0):
    v = np.ascontiguousarray(v, dtype=np.float32)
    out = np.empty_like(v)
    assert lib().oracle_mapoverlap1d(stencil, _p(v), _p(out), v.size, d, boundary, neutral) == 0
    return out


def gauss5_weights() -> np.ndarray:
    w = np.empty(25, dtype=np.float32)
    lib().oracle_gauss5_weights(_p(w))
    return w.reshape(5, 5)


AP_MANHATTAN, AP_DOT, AP_DOT_F64 = 0, 1, 2


def allpairs(fn: int, a: np.ndarray, b: np.ndarray) -> np.ndarray:
    """C[i][j] = A_i (+) B_j; rows of a (n x d) and b (m x d)."""
    a = np.ascontiguousarray(a, dtype=np.float32)
    b = np.ascontiguousarray(b, dtype=np.float32)
    n, d = a.shape
    m = b.shape[0]
    c = np.empty((n, m), dtype=np.float64 if fn == AP_DOT_F64 else np.float32)
    L = lib()
    L.oracle_allpairs.argtypes = [C.c_int, C.c_void_p, C.c_void_p, C.c_void_p, C.c_size_t, C.c_size_t, C.c_size_t]
    L.oracle_allpairs.restype = C.c_int
    assert L.oracle_allpairs(fn, _p(a), _p(b), _p(c), n, m, d) == 0
    return c


def block_range(n: int, G: int, g: int):
    lo, hi = C.c_size_t(), C.c_size_t()
    lib().oracle_block_range(n, G, g, C.byref(lo), C.byref(hi))
    return lo.value, hi.value


def overlap_range(n: int, G: int, g: int, d: int):
    lo, hi = C.c_size_t(), C.c_size_t()
    lib().oracle_overlap_range(n, G, g, d, C.byref(lo), C.byref(hi))
    return lo.value, hi.value


def siddon(p0, p1, N: int):
    p0 = np.ascontiguousarray(p0, dtype=np.float32)
    p1 = np.ascontiguousarray(p1, dtype=np.float32)
    cap = 6 * N + 8
    vox = np.empty(cap, dtype=np.int64)
    ln = np.empty(cap, dtype=np.float64)
    k = lib().oracle_siddon(_p(p0), _p(p1), N, _p(vox), _p(ln), cap)
    return vox[:k].copy(), ln[:k].copy()


def lmosem(events: np.ndarray, N: int, f: np.ndarray):
    """Returns (c, f_new, n_hit, visits) — c and f_new in float64."""
    events = np.ascontiguousarray(events, dtype=np.float32)
    f = np.ascontiguousarray(f, dtype=np.float32).reshape(-1)
    c = np.empty(N ** 3, dtype=np.float64)
    fn = np.empty(N ** 3, dtype=np.float64)
    vis = C.c_uint64()
    nhit = lib().oracle_lmosem(_p(events), events.shape[0], N, _p(f), _p(c), _p(fn), C.byref(vis))
    return c, fn, int(nhit), int(vis.value)
