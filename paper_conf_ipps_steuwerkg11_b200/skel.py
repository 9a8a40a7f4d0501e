"""Thin Python binding of libskel's C-ABI (include/skel.h): argument
marshalling only.  Every step of every skeleton runs in libskel's kernels;
there is no Python or CPU fallback -- if libskel.so is missing or no CUDA
device is usable, calls raise.

Names follow the paper (SkelCL, IPDPS 2011): Context ~ SkelCL::init
(P:L196), Vector (§III-A), Map/Zip/Reduce/Scan (§III-B), Arguments
(§III-C), distributions single/block/copy and setDistribution (§III-D,
Listing 4), mark_device_modified ~ dataOnDevicesModified.
"""
from __future__ import annotations

import ctypes
import os
from pathlib import Path

import numpy as np

LIB_PATH = Path(__file__).resolve().parent / "libskel.so"

SINGLE, BLOCK, COPY = 0, 1, 2
DIST_NAMES = {SINGLE: "single", BLOCK: "block", COPY: "copy"}
COMBINE_NONE, COMBINE_ADD, COMBINE_MIN, COMBINE_MAX, COMBINE_PROD = 0, 1, 2, 3, 4
ARG_SCALAR, ARG_VECTOR = 0, 1
XCHG_NAMES = ["none", "scatter", "broadcast", "gather", "allgather", "local_slice", "reduce_scatter",
              "keep_root", "reduce", "allreduce"]

_DT = {np.dtype(np.float32): 1, np.dtype(np.float64): 2, np.dtype(np.int32): 3, np.dtype(np.uint32): 4,
       np.dtype(np.int64): 5, np.dtype(np.uint64): 6}

STATUS = {0: "SKEL_OK", 1: "SKEL_ERR_ARG", 2: "SKEL_ERR_SIZE", 3: "SKEL_ERR_TYPE", 4: "SKEL_ERR_COMPILE",
          5: "SKEL_ERR_CUDA", 6: "SKEL_ERR_NCCL", 7: "SKEL_ERR_OOM", 8: "SKEL_ERR_STATE"}


class SkelError(RuntimeError):
    def __init__(self, status: int, msg: str):
        super().__init__(f"{STATUS.get(status, status)}: {msg}")
        self.status = status
        self.name = STATUS.get(status, str(status))
        self.msg = msg


class Stats(ctypes.Structure):
    _fields_ = [("h2d_bytes", ctypes.c_uint64), ("d2h_bytes", ctypes.c_uint64),
                ("h2d_copies", ctypes.c_uint64), ("d2h_copies", ctypes.c_uint64),
                ("d2d_bytes", ctypes.c_uint64), ("nccl_bytes", ctypes.c_uint64),
                ("kernel_launches", ctypes.c_uint64), ("compile_mem_hits", ctypes.c_uint64),
                ("compile_disk_hits", ctypes.c_uint64), ("compile_misses", ctypes.c_uint64),
                ("compile_ms", ctypes.c_double), ("disk_load_ms", ctypes.c_double),
                ("scan_coop_fallbacks", ctypes.c_uint64), ("vmm_allocs", ctypes.c_uint64),
                ("mc_binds", ctypes.c_uint64), ("multimem_launches", ctypes.c_uint64),
                ("xdev_reduces", ctypes.c_uint64)]

    def asdict(self):
        return {k: getattr(self, k) for k, _ in self._fields_}


class Arg(ctypes.Structure):
    _fields_ = [("kind", ctypes.c_int), ("data", ctypes.c_void_p), ("size", ctypes.c_size_t),
                ("vec", ctypes.c_void_p)]


_lib = None


def lib() -> ctypes.CDLL:
    """Load libskel.so (built in-tree by __graft_entry__.build())."""
    global _lib
    if _lib is None:
        if not LIB_PATH.exists():
            raise ImportError(f"{LIB_PATH} is not built: run `python -c 'import __graft_entry__ as g; g.build()'`")
        L = ctypes.CDLL(str(LIB_PATH))
        P, S, I = ctypes.c_void_p, ctypes.c_size_t, ctypes.c_int
        PP = ctypes.POINTER(ctypes.c_void_p)
        sig = {
            "skel_init": [I, PP], "skel_get_unique_id": [P], "skel_init_rank": [I, I, I, P, PP],
            "skel_finalize": [P], "skel_num_devices": [P, ctypes.POINTER(I), ctypes.POINTER(I)],
            "skel_get_stream": [P, I, PP], "skel_set_block_size": [P, I], "skel_set_cache_dir": [P, ctypes.c_char_p],
            "skel_clear_kernel_cache": [P], "skel_sync": [P], "skel_get_stats": [P, ctypes.POINTER(Stats)],
            "skel_reset_stats": [P],
            "skel_vector_create": [P, S, S, PP], "skel_vector_destroy": [P], "skel_vector_set_dtype": [P, I],
            "skel_vector_size": [P, ctypes.POINTER(S), ctypes.POINTER(S)], "skel_vector_upload": [P, P, S],
            "skel_vector_download": [P, P, S], "skel_vector_download_part": [P, S, P, S], "skel_vector_download_part_async": [P, S, P, S], "skel_vector_upload_part": [P, S, P, S], "skel_vector_host_ptr": [P, PP],
            "skel_vector_mark_host_modified": [P], "skel_vector_fill": [P, P], "skel_vector_fill_dist": [P, I, P],
            "skel_vector_set_distribution": [P, I, I], "skel_vector_get_distribution": [P, ctypes.POINTER(I)],
            "skel_vector_set_distribution_fn": [P, I, ctypes.c_char_p],
            "skel_vector_mark_device_modified": [P],
            "skel_vector_part": [P, I, ctypes.POINTER(S), ctypes.POINTER(S)],
            "skel_vector_device_ptr": [P, I, PP, ctypes.POINTER(S)],
            "skel_map": [P, ctypes.c_char_p, P, P, P, I], "skel_zip": [P, ctypes.c_char_p, P, P, P, P, I],
            "skel_map_index": [P, ctypes.c_char_p, S, P, P, I],
            "skel_map_lanes": [P, ctypes.c_char_p, P, P, I, P, I],
            "skel_reduce": [P, ctypes.c_char_p, P, P, P, I],
            "skel_zip_combine": [P, ctypes.c_char_p, P, P, I, P, P, I], "skel_reduce_to": [P, ctypes.c_char_p, P, P, P, I],
            "skel_scan": [P, ctypes.c_char_p, P, P, P, P, I], "skel_prepare": [P, ctypes.c_char_p, ctypes.c_char_p],
            "skel_entry_name": [ctypes.c_char_p, ctypes.c_char_p, S],
            "skel_compile_check": [ctypes.c_char_p, ctypes.c_char_p, I, ctypes.c_char_p, S, ctypes.POINTER(S)],
            "skel_plan_part": [S, I, I, ctypes.POINTER(S), ctypes.POINTER(S)],
            "skel_plan_exchange": [I, I, I, ctypes.POINTER(I)],
            "skel_capture_begin": [P], "skel_capture_end": [P, PP], "skel_graph_launch": [P],
            "skel_graph_destroy": [P],
        }
        for name, argt in sig.items():
            f = getattr(L, name)
            f.argtypes = argt
            f.restype = ctypes.c_int
        L.skel_last_error.argtypes = [P]
        L.skel_last_error.restype = ctypes.c_char_p
        L.skel_status_string.argtypes = [I]
        L.skel_status_string.restype = ctypes.c_char_p
        _lib = L
    return _lib


def _check(st: int, ctx=None):
    if st != 0:
        msg = lib().skel_last_error(ctx)
        raise SkelError(st, (msg or b"").decode(errors="replace"))


# ---------------------------------------------------------------------------
# pure host logic
# ---------------------------------------------------------------------------
def entry_name(src: str) -> str:
    buf = ctypes.create_string_buffer(256)
    _check(lib().skel_entry_name(src.encode(), buf, len(buf)))
    return buf.value.decode()


def compile_check(kind: str, src: str, fmad: bool = False) -> tuple[int, str, int]:
    """NVRTC-compile without a device: (status, log, cubin bytes)."""
    log = ctypes.create_string_buffer(1 << 16)
    sz = ctypes.c_size_t()
    st = lib().skel_compile_check(kind.encode(), src.encode(), int(fmad), log, len(log), ctypes.byref(sz))
    return st, log.value.decode(errors="replace"), sz.value


def plan_part(n: int, D: int, k: int) -> tuple[int, int]:
    lo, hi = ctypes.c_size_t(), ctypes.c_size_t()
    _check(lib().skel_plan_part(n, D, k, ctypes.byref(lo), ctypes.byref(hi)))
    return lo.value, hi.value


def plan_exchange(src: int, dst: int, combine: int = COMBINE_NONE) -> str:
    x = ctypes.c_int()
    _check(lib().skel_plan_exchange(src, dst, combine, ctypes.byref(x)))
    return XCHG_NAMES[x.value]


def unique_id() -> bytes:
    buf = ctypes.create_string_buffer(128)
    _check(lib().skel_get_unique_id(buf))
    return buf.raw


# ---------------------------------------------------------------------------
# context / vectors / skeletons
# ---------------------------------------------------------------------------
class Context:
    """SkelCL::init(): D logical devices in this process (num_devices), or
    one logical device per process (rank/world, NCCL exchanges)."""

    def __init__(self, num_devices: int = -1, *, rank: int | None = None, world: int | None = None,
                 device: int | None = None, nccl_id: bytes | None = None):
        self._h = ctypes.c_void_p()
        if rank is None:
            _check(lib().skel_init(num_devices, ctypes.byref(self._h)))
        else:
            idb = ctypes.create_string_buffer(nccl_id, 128) if nccl_id else None
            _check(lib().skel_init_rank(rank, world, rank if device is None else device, idb,
                                        ctypes.byref(self._h)))
        D, L = ctypes.c_int(), ctypes.c_int()
        _check(lib().skel_num_devices(self._h, ctypes.byref(D), ctypes.byref(L)), self._h)
        self.D, self.L = D.value, L.value
        self.rank = rank

    # -- lifecycle
    def close(self):
        if self._h:
            lib().skel_finalize(self._h)
            self._h = ctypes.c_void_p()

    def __enter__(self):
        return self

    def __exit__(self, *exc):
        self.close()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    @property
    def handle(self):
        return self._h

    def sync(self):
        _check(lib().skel_sync(self._h), self._h)

    def stats(self) -> dict:
        s = Stats()
        _check(lib().skel_get_stats(self._h, ctypes.byref(s)), self._h)
        return s.asdict()

    def reset_stats(self):
        _check(lib().skel_reset_stats(self._h), self._h)

    def stream(self, local_index: int = 0) -> int:
        p = ctypes.c_void_p()
        _check(lib().skel_get_stream(self._h, local_index, ctypes.byref(p)), self._h)
        return p.value or 0

    def set_block_size(self, threads: int):
        _check(lib().skel_set_block_size(self._h, threads), self._h)

    def set_cache_dir(self, path: str | None):
        _check(lib().skel_set_cache_dir(self._h, None if path is None else path.encode()), self._h)

    def clear_kernel_cache(self):
        _check(lib().skel_clear_kernel_cache(self._h), self._h)

    def prepare(self, kind: str, src: str):
        _check(lib().skel_prepare(self._h, kind.encode(), src.encode()), self._h)

    # -- CUDA graphs
    def capture_begin(self):
        _check(lib().skel_capture_begin(self._h), self._h)

    def capture_end(self) -> "Graph":
        g = ctypes.c_void_p()
        _check(lib().skel_capture_end(self._h, ctypes.byref(g)), self._h)
        return Graph(self, g)

    def capture(self, fn) -> "Graph":
        """Record the device work of fn() into a replayable graph."""
        self.capture_begin()
        try:
            fn()
        except BaseException:
            try:
                self.capture_end().destroy()
            except SkelError:
                pass
            raise
        return self.capture_end()

    # -- vectors
    def vector(self, data=None, *, n: int | None = None, dtype=None) -> "Vector":
        if data is not None:
            arr = np.ascontiguousarray(data)
            v = Vector(self, arr.size, arr.dtype)
            v.upload(arr)
            return v
        return Vector(self, int(n), np.dtype(dtype))

    # -- skeletons
    def _args(self, args):
        arr = (Arg * max(1, len(args)))()
        keep = []
        for i, a in enumerate(args):
            if isinstance(a, Vector):
                arr[i].kind, arr[i].vec = ARG_VECTOR, a._h.value
            else:
                b = np.ascontiguousarray(np.asarray(a).reshape(1))
                keep.append(b)
                arr[i].kind, arr[i].data, arr[i].size = ARG_SCALAR, b.ctypes.data, b.dtype.itemsize
        return arr, keep

    def map(self, src: str, vin: "Vector", vout: "Vector | None" = None, args=()):
        """eq. (1): vout[i] = f(vin[i], args...); vout=None for a void (side-effect) Map."""
        a, keep = self._args(args)
        _check(lib().skel_map(self._h, src.encode(), vin._h, vout._h if vout is not None else None, a, len(args)), self._h)
        return vout

    def map_index(self, src: str, n: int, vout: "Vector | None" = None, args=()):
        """NEXT-4: out[i] = f(i, args...) for i in [0, n), no input vector."""
        a, keep = self._args(args)
        _check(lib().skel_map_index(self._h, src.encode(), n, vout._h if vout is not None else None, a, len(args)),
               self._h)
        return vout

    def map_lanes(self, src: str, vin: "Vector", vout: "Vector | None" = None, lanes: int = 1, args=()):
        """Map with `lanes` threads per element: f(x, lane, lanes, args...)."""
        a, keep = self._args(args)
        _check(lib().skel_map_lanes(self._h, src.encode(), vin._h, vout._h if vout is not None else None, lanes,
                                    a, len(args)), self._h)
        return vout

    def zip(self, src: str, va: "Vector", vb: "Vector", vout: "Vector", args=()):
        """eq. (2): vout[i] = f(va[i], vb[i], args...)."""
        a, keep = self._args(args)
        _check(lib().skel_zip(self._h, src.encode(), va._h, vb._h, vout._h, a, len(args)), self._h)
        return vout

    def zip_combine(self, src: str, va: "Vector", vb: "Vector", combine: int, vout: "Vector", args=()):
        """vb.set_distribution(BLOCK, combine); vout = zip(va, vb); vout -> COPY, fused (NEXT-1)."""
        a, keep = self._args(args)
        _check(lib().skel_zip_combine(self._h, src.encode(), va._h, vb._h, combine, vout._h, a, len(args)), self._h)
        return vout

    def reduce(self, src: str, vin: "Vector", args=()):
        """eq. (3): the fold of vin, returned to the host (Scalar::getValue)."""
        a, keep = self._args(args)
        out = np.zeros(1, dtype=vin.dtype)
        _check(lib().skel_reduce(self._h, src.encode(), vin._h, out.ctypes.data, a, len(args)), self._h)
        return out[0]

    def reduce_to(self, src: str, vin: "Vector", result: "Vector", args=()):
        a, keep = self._args(args)
        _check(lib().skel_reduce_to(self._h, src.encode(), vin._h, result._h, a, len(args)), self._h)
        return result

    def scan(self, src: str, vin: "Vector", vout: "Vector", identity, args=()):
        """eq. (4): exclusive scan with the given identity."""
        a, keep = self._args(args)
        idv = np.ascontiguousarray(np.asarray(identity, dtype=vin.dtype).reshape(1))
        _check(lib().skel_scan(self._h, src.encode(), vin._h, vout._h, idv.ctypes.data, a, len(args)), self._h)
        return vout


class Graph:
    """A captured skeleton sequence (CUDA graph) that can be replayed."""

    def __init__(self, ctx: Context, h):
        self.ctx, self._h = ctx, h

    def launch(self):
        _check(lib().skel_graph_launch(self._h), self.ctx._h)

    def destroy(self):
        if self._h and self._h.value:
            lib().skel_graph_destroy(self._h)
        self._h = ctypes.c_void_p()

    def __del__(self):
        try:
            self.destroy()
        except Exception:
            pass


class Vector:
    """Vector<T> (§III-A): host mirror + per-device storage, lazy coherence."""

    def __init__(self, ctx: Context, n: int, dtype):
        self.ctx = ctx
        self.dtype = np.dtype(dtype)
        self._h = ctypes.c_void_p()
        _check(lib().skel_vector_create(ctx._h, n, self.dtype.itemsize, ctypes.byref(self._h)), ctx._h)
        if self.dtype in _DT:
            _check(lib().skel_vector_set_dtype(self._h, _DT[self.dtype]), ctx._h)

    def destroy(self):
        if self._h and self.ctx._h:
            lib().skel_vector_destroy(self._h)
        self._h = ctypes.c_void_p()

    def __del__(self):
        try:
            self.destroy()
        except Exception:
            pass

    @property
    def n(self) -> int:
        n, es = ctypes.c_size_t(), ctypes.c_size_t()
        _check(lib().skel_vector_size(self._h, ctypes.byref(n), ctypes.byref(es)), self.ctx._h)
        return n.value

    def __len__(self):
        return self.n

    def upload(self, arr):
        a = np.ascontiguousarray(arr, dtype=self.dtype).reshape(-1)
        _check(lib().skel_vector_upload(self._h, a.ctypes.data, a.size), self.ctx._h)
        return self

    def upload_part(self, lo: int, arr):
        """Host data for elements [lo, lo + len(arr)) (rank-local mirror in rank mode)."""
        a = np.ascontiguousarray(arr, dtype=self.dtype).reshape(-1)
        _check(lib().skel_vector_upload_part(self._h, lo, a.ctypes.data, a.size), self.ctx._h)
        return self

    def download(self) -> np.ndarray:
        out = np.empty(self.n, dtype=self.dtype)
        _check(lib().skel_vector_download(self._h, out.ctypes.data, out.size), self.ctx._h)
        return out

    def download_part(self, lo: int, out: np.ndarray) -> np.ndarray:
        """Elements [lo, lo + out.size) into `out` (straight from the devices
        holding them; pass pinned memory for full-rate copies)."""
        assert out.dtype == self.dtype and out.flags["C_CONTIGUOUS"]
        _check(lib().skel_vector_download_part(self._h, lo, out.ctypes.data, out.size), self.ctx._h)
        return out

    def download_part_async(self, lo: int, out: np.ndarray) -> np.ndarray:
        """As download_part, without waiting: `out` (pinned memory) is filled by the
        time of the next ctx.sync()."""
        assert out.dtype == self.dtype and out.flags["C_CONTIGUOUS"]
        _check(lib().skel_vector_download_part_async(self._h, lo, out.ctypes.data, out.size), self.ctx._h)
        return out

    def host_view(self) -> np.ndarray:
        """numpy view of the pinned host mirror (valid until the vector changes size)."""
        p = ctypes.c_void_p()
        _check(lib().skel_vector_host_ptr(self._h, ctypes.byref(p)), self.ctx._h)
        n = self.n
        buf = (ctypes.c_char * (n * self.dtype.itemsize)).from_address(p.value)
        return np.frombuffer(buf, dtype=self.dtype, count=n)

    def mark_host_modified(self):
        _check(lib().skel_vector_mark_host_modified(self._h), self.ctx._h)

    def fill(self, value):
        b = np.ascontiguousarray(np.asarray(value, dtype=self.dtype).reshape(1))
        _check(lib().skel_vector_fill(self._h, b.ctypes.data), self.ctx._h)
        return self

    def fill_dist(self, dist: int, value):
        """Discard contents, take distribution `dist` (no exchange), fill with value."""
        b = np.ascontiguousarray(np.asarray(value, dtype=self.dtype).reshape(1))
        _check(lib().skel_vector_fill_dist(self._h, dist, b.ctypes.data), self.ctx._h)
        return self

    def set_distribution(self, dist: int, combine: "int | str" = COMBINE_NONE):
        """combine: a built-in skel_combine, or source text of a user function
        T f(T, T) (skel_vector_set_distribution_fn, NEXT-2)."""
        if isinstance(combine, str):
            _check(lib().skel_vector_set_distribution_fn(self._h, dist, combine.encode()), self.ctx._h)
        else:
            _check(lib().skel_vector_set_distribution(self._h, dist, combine), self.ctx._h)
        return self

    @property
    def distribution(self) -> int:
        d = ctypes.c_int()
        _check(lib().skel_vector_get_distribution(self._h, ctypes.byref(d)), self.ctx._h)
        return d.value

    def mark_device_modified(self):
        _check(lib().skel_vector_mark_device_modified(self._h), self.ctx._h)

    def part(self, d: int) -> tuple[int, int]:
        lo, hi = ctypes.c_size_t(), ctypes.c_size_t()
        _check(lib().skel_vector_part(self._h, d, ctypes.byref(lo), ctypes.byref(hi)), self.ctx._h)
        return lo.value, hi.value

    def device_ptr(self, local_index: int = 0) -> tuple[int, int]:
        p, c = ctypes.c_void_p(), ctypes.c_size_t()
        _check(lib().skel_vector_device_ptr(self._h, local_index, ctypes.byref(p), ctypes.byref(c)), self.ctx._h)
        return p.value or 0, c.value
