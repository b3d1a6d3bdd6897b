"""Thin Python binding of libskl.so (include/skl.h) — argument marshalling only.

Every skeleton runs in the library's NVRTC-compiled sm_100a kernels; nothing in
this module computes.  If libskl.so is missing the import fails loudly: there
is no CPU fallback.

    ctx = Context()                                   # SkelCL::init()
    neg = Map(ctx, "float func(float x){ return -x;}", F32, F32)
    out = neg(Vector.from_numpy(ctx, x))
    out.to_numpy()                                    # implicit download
"""
from __future__ import annotations

import ctypes as C
import os
from typing import Optional, Sequence

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "libskl.so")

# element types (skl.h)
VOID, U8, I8, I32, U32, F32, F64, F32X2, I64, U64, I16, U16 = range(12)
PTR = 0x1000
# distributions
DIST_NONE, SINGLE, COPY, BLOCK, OVERLAP = range(5)
NEUTRAL, NEAREST = 0, 1
READ, WRITE, RW = 1, 2, 3
ARG_SCALAR, ARG_CONT = 1, 2

ERRORS = {-1: "INVALID_ARG", -2: "TYPE", -3: "SIZE_MISMATCH", -4: "EMPTY", -5: "COMPILE",
          -6: "OUT_OF_RANGE", -7: "DISTRIBUTION", -8: "OOM", -9: "CUDA", -10: "NCCL",
          -11: "UNSUPPORTED"}

_NP = {U8: np.uint8, I8: np.int8, I32: np.int32, U32: np.uint32, F32: np.float32, F64: np.float64,
       I64: np.int64, U64: np.uint64, I16: np.int16, U16: np.uint16, F32X2: np.float32}


class SklError(RuntimeError):
    def __init__(self, code: int, msg: str):
        super().__init__(f"SKL_ERR_{ERRORS.get(code, code)}: {msg}")
        self.code = code
        self.name = ERRORS.get(code, str(code))


class _Arg(C.Structure):
    _fields_ = [("kind", C.c_int), ("mode", C.c_int), ("value", C.c_void_p), ("bytes", C.c_size_t),
                ("cont", C.c_void_p)]


_lib = None


def lib():
    """Load libskl.so (raises if it was not built: no fallback)."""
    global _lib
    if _lib is not None:
        return _lib
    if not os.path.exists(_SO):
        raise ImportError(f"{_SO} not built: run `python -m paper_conf_pact_steuwerg13_b200.build` "
                          "(there is no CPU fallback)")
    L = C.CDLL(_SO)
    vp, sz, i, pp = C.c_void_p, C.c_size_t, C.c_int, C.POINTER(C.c_void_p)
    sig = {
        "skl_init": [i, vp, pp], "skl_init_dist": [i, i, i, vp, pp], "skl_init_offline": [pp],
        "skl_nccl_unique_id": [vp], "skl_finalize": [vp],
        "skl_num_devices": [vp, C.POINTER(i), C.POINTER(i), C.POINTER(i)],
        "skl_set_stream": [vp, i, vp], "skl_get_stream": [vp, i, pp], "skl_sync": [vp],
        "skl_set_allocator": [vp, vp, vp, vp],
        "skl_set_option": [vp, C.c_char_p, C.c_longlong],
        "skl_get_counter": [vp, C.c_char_p, C.POINTER(C.c_longlong)],
        "skl_type_struct": [vp, C.c_char_p, C.c_char_p, sz, sz, C.POINTER(i)],
        "skl_type_size": [vp, i, C.POINTER(sz)],
        "skl_vector_create": [vp, i, sz, pp], "skl_matrix_create": [vp, i, sz, sz, pp],
        "skl_cont_destroy": [vp], "skl_cont_info": [vp, C.POINTER(i), C.POINTER(sz), C.POINTER(sz), C.POINTER(i)],
        "skl_copy_in": [vp, vp, sz], "skl_copy_out": [vp, vp, sz],
        "skl_copy_out_part": [vp, i, vp, sz, C.POINTER(sz), C.POINTER(sz)],
        "skl_host_data": [vp, i, pp], "skl_fill": [vp, vp],
        "skl_set_distribution": [vp, i, i, vp], "skl_get_distribution": [vp, C.POINTER(i), C.POINTER(i)],
        "skl_local_part": [vp, i, pp, C.POINTER(sz), C.POINTER(sz)],
        "skl_map_create": [vp, C.c_char_p, C.c_char_p, i, i, C.POINTER(i), i, pp],
        "skl_zip_create": [vp, C.c_char_p, C.c_char_p, i, i, i, C.POINTER(i), i, pp],
        "skl_reduce_create": [vp, C.c_char_p, C.c_char_p, i, pp],
        "skl_scan_create": [vp, C.c_char_p, C.c_char_p, i, pp],
        "skl_mapoverlap_create": [vp, C.c_char_p, C.c_char_p, i, i, i, i, vp, pp],
        "skl_skel_destroy": [vp],
        "skl_map_run": [vp, vp, pp, C.POINTER(_Arg), i],
        "skl_zip_run": [vp, vp, vp, pp, C.POINTER(_Arg), i],
        "skl_reduce_run": [vp, vp, pp], "skl_scan_run": [vp, vp, pp], "skl_mapoverlap_run": [vp, vp, pp],
        "skl_scalar_get": [vp, vp, sz],
        "skl_skel_cubin": [vp, vp, sz, C.POINTER(sz)], "skl_skel_source": [vp, C.c_char_p, sz, C.POINTER(sz)],
        "skl_mapoverlap_bounds": [vp, C.POINTER(i)],
        "skl_allpairs_create": [vp, C.c_char_p, C.c_char_p, i, i, pp],
        "skl_allpairs_zr_create": [vp, C.c_char_p, C.c_char_p, C.c_char_p, C.c_char_p, i, i, pp],
        "skl_allpairs_run": [vp, vp, vp, pp],
        "skl_capture_begin": [vp], "skl_capture_end": [vp, pp], "skl_graph_launch": [vp],
        "skl_graph_destroy": [vp],
        "skl_plan_range": [sz, i, i, i, i, i, C.POINTER(sz), C.POINTER(sz)],
        "skl_plan_transfers": [sz, i, i, i, i, i, C.POINTER(C.c_int64), sz, C.POINTER(sz)],
    }
    for name, args in sig.items():
        f = getattr(L, name)
        f.argtypes = args
        f.restype = C.c_int
    L.skl_last_error.restype = C.c_char_p
    L.skl_last_error.argtypes = []
    _lib = L
    return L


def check(rc: int):
    if rc != 0:
        msg = lib().skl_last_error()
        raise SklError(rc, msg.decode(errors="replace") if msg else "")


def exported_symbols() -> list:
    return [n for n in dir(lib()) if n.startswith("skl_")]


_ALLOC_FN = C.CFUNCTYPE(C.c_void_p, C.c_size_t, C.c_int, C.c_void_p, C.c_void_p)
_FREE_FN = C.CFUNCTYPE(None, C.c_void_p, C.c_int, C.c_void_p, C.c_void_p)


# ---------------------------------------------------------------- context
class Context:
    """SkelCL::init().  ndev logical devices over `devices` (CUDA ordinals)."""

    def __init__(self, ndev: int = 0, devices: Optional[Sequence[int]] = None, _handle=None):
        self._h = C.c_void_p()
        if _handle is not None:
            self._h = _handle
        else:
            arr = (C.c_int * len(devices))(*devices) if devices else None
            if devices and ndev == 0:
                ndev = len(devices)
            check(lib().skl_init(ndev, arr, C.byref(self._h)))
        self._live = True
        self._types = {}

    @classmethod
    def dist(cls, rank: int, world: int, device: int, nccl_id: bytes) -> "Context":
        h = C.c_void_p()
        buf = C.create_string_buffer(nccl_id, 128) if nccl_id is not None else None
        check(lib().skl_init_dist(rank, world, device, buf, C.byref(h)))
        return cls(_handle=h)

    @classmethod
    def offline(cls) -> "Context":
        h = C.c_void_p()
        check(lib().skl_init_offline(C.byref(h)))
        return cls(_handle=h)

    @staticmethod
    def nccl_unique_id() -> bytes:
        buf = C.create_string_buffer(128)
        check(lib().skl_nccl_unique_id(buf))
        return buf.raw

    @property
    def handle(self):
        return self._h

    def devices(self):
        n, f, l = C.c_int(), C.c_int(), C.c_int()
        check(lib().skl_num_devices(self._h, C.byref(n), C.byref(f), C.byref(l)))
        return n.value, f.value, l.value

    @property
    def ndev(self) -> int:
        return self.devices()[0]

    def set_stream(self, g: int, stream: int):
        check(lib().skl_set_stream(self._h, g, C.c_void_p(stream) if stream else None))

    def stream(self, g: int) -> int:
        s = C.c_void_p()
        check(lib().skl_get_stream(self._h, g, C.byref(s)))
        return s.value or 0

    def sync(self):
        check(lib().skl_sync(self._h))

    def use_torch_allocator(self):
        """Route the library's device memory through torch's caching allocator
        (skl_set_allocator; PyTorch as the device-memory plumbing).  Call before
        creating containers or skeletons."""
        import torch

        def _alloc(nbytes, dev, stream, _user):
            try:
                return torch.cuda.caching_allocator_alloc(nbytes, dev, stream or 0)
            except Exception:   # noqa: BLE001 - the library reports SKL_ERR_OOM
                return None

        def _free(ptr, _dev, _stream, _user):
            torch.cuda.caching_allocator_delete(ptr)

        self._alloc_cb = (_ALLOC_FN(_alloc), _FREE_FN(_free))   # kept alive with the context
        check(lib().skl_set_allocator(self._h, C.cast(self._alloc_cb[0], C.c_void_p),
                                      C.cast(self._alloc_cb[1], C.c_void_p), None))

    def set_option(self, key: str, value: int):
        check(lib().skl_set_option(self._h, key.encode(), value))

    def counter(self, key: str) -> int:
        v = C.c_longlong()
        check(lib().skl_get_counter(self._h, key.encode(), C.byref(v)))
        return v.value

    def struct_type(self, name: str, decl: str, size: int, align: int = 4) -> int:
        t = C.c_int()
        check(lib().skl_type_struct(self._h, name.encode(), decl.encode(), size, align, C.byref(t)))
        return t.value

    def capture(self, fn) -> "Graph":
        """Record fn() (skeleton calls on this context) as a CUDA graph."""
        check(lib().skl_capture_begin(self._h))
        try:
            fn()
        except BaseException:
            h = C.c_void_p()
            lib().skl_capture_end(self._h, C.byref(h))
            if h.value:
                lib().skl_graph_destroy(h)
            raise
        h = C.c_void_p()
        check(lib().skl_capture_end(self._h, C.byref(h)))
        return Graph(self, h)

    def finalize(self):
        if self._live:
            check(lib().skl_finalize(self._h))
            self._live = False

    def __enter__(self):
        return self

    def __exit__(self, *a):
        self.finalize()


class Graph:
    """A recorded sequence of skeleton calls (skl_capture_begin/end)."""

    def __init__(self, ctx: Context, h):
        self.ctx = ctx
        self._h = h

    def launch(self):
        check(lib().skl_graph_launch(self._h))

    def destroy(self):
        if self._h:
            check(lib().skl_graph_destroy(self._h))
            self._h = None


# ---------------------------------------------------------------- containers
class Container:
    """Vector<T> / Matrix<T>."""

    def __init__(self, ctx: Context, handle, dtype: int):
        self.ctx = ctx
        self._h = handle
        self.dtype = dtype

    @property
    def handle(self):
        return self._h

    def info(self):
        t, r, c, m = C.c_int(), C.c_size_t(), C.c_size_t(), C.c_int()
        check(lib().skl_cont_info(self._h, C.byref(t), C.byref(r), C.byref(c), C.byref(m)))
        return t.value, r.value, c.value, bool(m.value)

    @property
    def shape(self):
        _, r, c, m = self.info()
        return (r, c) if m else (r,)

    def elem_size(self) -> int:
        s = C.c_size_t()
        check(lib().skl_type_size(self.ctx.handle, self.dtype, C.byref(s)))
        return s.value

    @property
    def nbytes(self) -> int:
        n = 1
        for s in self.shape:
            n *= s
        return n * self.elem_size()

    def copy_in(self, host: np.ndarray):
        host = np.ascontiguousarray(host)
        if host.nbytes != self.nbytes:
            raise SklError(-3, f"copy_in: {host.nbytes} bytes for a {self.nbytes}-byte container")
        check(lib().skl_copy_in(self._h, host.ctypes.data_as(C.c_void_p), host.nbytes))
        return self

    def copy_in_ptr(self, ptr: int, nbytes: int):
        check(lib().skl_copy_in(self._h, C.c_void_p(ptr), nbytes))

    def copy_out_ptr(self, ptr: int, nbytes: int):
        check(lib().skl_copy_out(self._h, C.c_void_p(ptr), nbytes))

    def to_numpy(self, np_dtype=None) -> np.ndarray:
        np_dtype = np_dtype or _NP.get(self.dtype, np.uint8)
        shape = self.shape
        if self.dtype == F32X2:
            shape = shape + (2,)
        out = np.empty(self.nbytes // np.dtype(np_dtype).itemsize, dtype=np_dtype)
        check(lib().skl_copy_out(self._h, out.ctypes.data_as(C.c_void_p), out.nbytes))
        if np_dtype == _NP.get(self.dtype) or self.dtype == F32X2:
            out = out.reshape(shape)
        return out

    def copy_out_part(self, g: int, host: np.ndarray):
        f, n = C.c_size_t(), C.c_size_t()
        check(lib().skl_copy_out_part(self._h, g, host.ctypes.data_as(C.c_void_p), host.nbytes,
                                      C.byref(f), C.byref(n)))
        return f.value, n.value

    def host_data(self, mode: int = RW) -> int:
        p = C.c_void_p()
        check(lib().skl_host_data(self._h, mode, C.byref(p)))
        return p.value

    def fill(self, value):
        v = np.array([value], dtype=_NP[self.dtype]) if not isinstance(value, np.ndarray) else value
        check(lib().skl_fill(self._h, v.ctypes.data_as(C.c_void_p)))
        return self

    def set_distribution(self, kind: int, arg: int = 0, combine: "Skeleton" = None):
        check(lib().skl_set_distribution(self._h, kind, arg, combine.handle if combine else None))
        return self

    def distribution(self):
        k, a = C.c_int(), C.c_int()
        check(lib().skl_get_distribution(self._h, C.byref(k), C.byref(a)))
        return k.value, a.value

    def local_part(self, g: int):
        p, f, n = C.c_void_p(), C.c_size_t(), C.c_size_t()
        check(lib().skl_local_part(self._h, g, C.byref(p), C.byref(f), C.byref(n)))
        return p.value, f.value, n.value

    def scalar(self, np_dtype=None):
        np_dtype = np_dtype or _NP[self.dtype]
        v = np.empty(self.nbytes // np.dtype(np_dtype).itemsize, dtype=np_dtype)
        check(lib().skl_scalar_get(self._h, v.ctypes.data_as(C.c_void_p), v.nbytes))
        return v[0] if v.size == 1 else v

    def destroy(self):
        if self._h:
            check(lib().skl_cont_destroy(self._h))
            self._h = None

    def __del__(self):
        # containers die with their Python object (device memory freed stream-
        # ordered); after Context.finalize() the library already freed them
        try:
            if self._h and self.ctx._live:
                lib().skl_cont_destroy(self._h)
                self._h = None
        except Exception:
            pass


class Vector(Container):
    def __init__(self, ctx: Context, dtype: int, n: int):
        h = C.c_void_p()
        check(lib().skl_vector_create(ctx.handle, dtype, n, C.byref(h)))
        super().__init__(ctx, h, dtype)

    @classmethod
    def from_numpy(cls, ctx: Context, a: np.ndarray, dtype: int = None) -> "Vector":
        dtype = dtype if dtype is not None else _from_np(a.dtype)
        n = a.shape[0] if a.ndim else 1
        v = cls(ctx, dtype, n)
        return v.copy_in(a)


class Matrix(Container):
    def __init__(self, ctx: Context, dtype: int, rows: int, cols: int):
        h = C.c_void_p()
        check(lib().skl_matrix_create(ctx.handle, dtype, rows, cols, C.byref(h)))
        super().__init__(ctx, h, dtype)

    @classmethod
    def from_numpy(cls, ctx: Context, a: np.ndarray, dtype: int = None) -> "Matrix":
        dtype = dtype if dtype is not None else _from_np(a.dtype)
        m = cls(ctx, dtype, a.shape[0], a.shape[1])
        return m.copy_in(a)


def _from_np(dt) -> int:
    for k, v in _NP.items():
        if k != F32X2 and np.dtype(v) == np.dtype(dt):
            return k
    raise SklError(-2, f"no SkelCL element type for numpy dtype {dt}")


def _wrap_out(ctx, handle, dtype):
    return Container(ctx, handle, dtype)


# ---------------------------------------------------------------- skeletons
class Skeleton:
    def __init__(self, ctx: Context, handle, tout: int):
        self.ctx = ctx
        self._h = handle
        self.tout = tout

    @property
    def handle(self):
        return self._h

    def cubin(self) -> bytes:
        n = C.c_size_t()
        check(lib().skl_skel_cubin(self._h, None, 0, C.byref(n)))
        buf = C.create_string_buffer(n.value)
        check(lib().skl_skel_cubin(self._h, buf, n.value, C.byref(n)))
        return buf.raw[: n.value]

    def source(self) -> str:
        n = C.c_size_t()
        check(lib().skl_skel_source(self._h, None, 0, C.byref(n)))
        buf = C.create_string_buffer(n.value)
        check(lib().skl_skel_source(self._h, buf, n.value, C.byref(n)))
        return buf.value.decode()

    def destroy(self):
        if self._h:
            check(lib().skl_skel_destroy(self._h))
            self._h = None

    @staticmethod
    def _extras(extra):
        arr = (_Arg * max(1, len(extra)))()
        keep = []
        for k, e in enumerate(extra):
            if isinstance(e, tuple) and isinstance(e[0], Container):
                arr[k].kind, arr[k].mode, arr[k].cont = ARG_CONT, e[1], e[0].handle
            elif isinstance(e, Container):
                arr[k].kind, arr[k].mode, arr[k].cont = ARG_CONT, READ, e.handle
            else:
                v = np.ascontiguousarray(e)
                keep.append(v)
                arr[k].kind, arr[k].value, arr[k].bytes = ARG_SCALAR, v.ctypes.data, v.nbytes
        return arr, keep


def _types(ts):
    ts = list(ts or [])
    return (C.c_int * max(1, len(ts)))(*ts), len(ts)


class Map(Skeleton):
    """map f [c1..cn] = [f(c1)..f(cn)]."""

    def __init__(self, ctx, src: str, tin: int, tout: int, extra: Sequence[int] = (), entry: str = None):
        h = C.c_void_p()
        xt, nx = _types(extra)
        check(lib().skl_map_create(ctx.handle, src.encode(), entry.encode() if entry else None, tin, tout,
                                   xt, nx, C.byref(h)))
        super().__init__(ctx, h, tout)

    def __call__(self, inp: Container, *extra, out: Container = None):
        o = C.c_void_p(out.handle.value if out is not None else None)
        arr, keep = self._extras(extra)
        check(lib().skl_map_run(self._h, inp.handle, C.byref(o), arr, len(extra)))
        if self.tout == VOID:
            return None
        return out if out is not None else _wrap_out(self.ctx, o, self.tout)


class Zip(Skeleton):
    """zip (+) [cl][cr] = [cl_i (+) cr_i]."""

    def __init__(self, ctx, src: str, tl: int, tr: int, tout: int, extra: Sequence[int] = (), entry=None):
        h = C.c_void_p()
        xt, nx = _types(extra)
        check(lib().skl_zip_create(ctx.handle, src.encode(), entry.encode() if entry else None, tl, tr, tout,
                                   xt, nx, C.byref(h)))
        super().__init__(ctx, h, tout)

    def __call__(self, left: Container, right: Container, *extra, out: Container = None):
        o = C.c_void_p(out.handle.value if out is not None else None)
        arr, keep = self._extras(extra)
        check(lib().skl_zip_run(self._h, left.handle, right.handle, C.byref(o), arr, len(extra)))
        if self.tout == VOID:
            return None
        return out if out is not None else _wrap_out(self.ctx, o, self.tout)


class Reduce(Skeleton):
    """red (+) [v1..vn] = v1 (+) ... (+) vn; returns a Scalar container."""

    def __init__(self, ctx, src: str, t: int, entry=None):
        h = C.c_void_p()
        check(lib().skl_reduce_create(ctx.handle, src.encode(), entry.encode() if entry else None, t, C.byref(h)))
        super().__init__(ctx, h, t)

    def __call__(self, inp: Container, out: Container = None) -> Container:
        o = C.c_void_p(out.handle.value if out is not None else None)
        check(lib().skl_reduce_run(self._h, inp.handle, C.byref(o)))
        return out if out is not None else _wrap_out(self.ctx, o, self.tout)


class Scan(Skeleton):
    """inclusive scan (+)."""

    def __init__(self, ctx, src: str, t: int, entry=None):
        h = C.c_void_p()
        check(lib().skl_scan_create(ctx.handle, src.encode(), entry.encode() if entry else None, t, C.byref(h)))
        super().__init__(ctx, h, t)

    def __call__(self, inp: Container, out: Container = None) -> Container:
        o = C.c_void_p(out.handle.value if out is not None else None)
        check(lib().skl_scan_run(self._h, inp.handle, C.byref(o)))
        return out if out is not None else _wrap_out(self.ctx, o, self.tout)


class MapOverlap(Skeleton):
    """mout[i,j] = f(window [-d,+d]^2) with get(p,dx,dy)."""

    def __init__(self, ctx, src: str, tin: int, tout: int, d: int, boundary: int = NEUTRAL,
                 neutral=0, entry=None):
        h = C.c_void_p()
        nv = np.array([neutral], dtype=_NP.get(tin, np.uint8))
        check(lib().skl_mapoverlap_create(ctx.handle, src.encode(), entry.encode() if entry else None, tin, tout,
                                          d, boundary, nv.ctypes.data_as(C.c_void_p), C.byref(h)))
        super().__init__(ctx, h, tout)

    def __call__(self, inp: Container, out: Container = None) -> Container:
        o = C.c_void_p(out.handle.value if out is not None else None)
        check(lib().skl_mapoverlap_run(self._h, inp.handle, C.byref(o)))
        return out if out is not None else _wrap_out(self.ctx, o, self.tout)

    @property
    def bounds_proven(self) -> bool:
        """get() offsets statically proven within [-d, d]."""
        v = C.c_int()
        check(lib().skl_mapoverlap_bounds(self._h, C.byref(v)))
        return bool(v.value)


class Allpairs(Skeleton):
    """allpairs(+)(A, B): C[i][j] = A_i (+) B_j over rows.

    Allpairs(ctx, "float f(const float* a, const float* b, int d){...}", F32, F32)
    Allpairs(ctx, zip_src, F32, F32, reduce=reduce_src)   # fold((+), zip((x), A_i, B_j))
    """

    def __init__(self, ctx, src: str, tin: int, tout: int, reduce: str = None, entry=None,
                 reduce_entry=None):
        h = C.c_void_p()
        if reduce is None:
            check(lib().skl_allpairs_create(ctx.handle, src.encode(), entry.encode() if entry else None,
                                            tin, tout, C.byref(h)))
        else:
            check(lib().skl_allpairs_zr_create(ctx.handle, src.encode(), entry.encode() if entry else None,
                                               reduce.encode(), reduce_entry.encode() if reduce_entry else None,
                                               tin, tout, C.byref(h)))
        super().__init__(ctx, h, tout)

    def __call__(self, a: Container, b: Container, out: Container = None) -> Container:
        o = C.c_void_p(out.handle.value if out is not None else None)
        check(lib().skl_allpairs_run(self._h, a.handle, b.handle, C.byref(o)))
        return out if out is not None else _wrap_out(self.ctx, o, self.tout)


# ---------------------------------------------------------------- host-only planning
def plan_range(units: int, G: int, kind: int, arg: int, g: int, with_halo: bool):
    lo, hi = C.c_size_t(), C.c_size_t()
    check(lib().skl_plan_range(units, G, kind, arg, g, int(with_halo), C.byref(lo), C.byref(hi)))
    return lo.value, hi.value


def plan_transfers(units: int, G: int, from_kind: int, from_arg: int, to_kind: int, to_arg: int):
    n = C.c_size_t()
    check(lib().skl_plan_transfers(units, G, from_kind, from_arg, to_kind, to_arg, None, 0, C.byref(n)))
    buf = (C.c_int64 * max(1, 5 * n.value))()
    check(lib().skl_plan_transfers(units, G, from_kind, from_arg, to_kind, to_arg, buf, n.value, C.byref(n)))
    return [tuple(buf[5 * i: 5 * i + 5]) for i in range(n.value)]
