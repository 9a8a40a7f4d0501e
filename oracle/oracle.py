"""Python face of the CPU oracle -- TEST INFRASTRUCTURE ONLY.

Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline /
`--impl reference` legs may import this module.  The product package
(paper_conf_ipps_steuwerkg11_b200) never imports it, and it never imports the
product package: the two share only the seeded generators of skel_inputs/.

Two native pieces, both plain sequential C/C++ built with
``-O2 -ffp-contract=off -fno-fast-math`` (reading R11):

* ``liboracle_core.so`` from oracle_core.c: Mandelbrot (eq. 5), Siddon
  compute_path, LM OSEM Listing 3, exact float sums/prefix sums;
* one ``.so`` per (user function source, skeleton): the user function text
  ("a plain string containing the function's source code")
  compiled by g++ together with the sequential skeleton loops of
  skel_oracle_impl.hpp (eqs. (1)-(4)).
"""
from __future__ import annotations

import ctypes
import hashlib
import os
import re
import subprocess
from pathlib import Path

import numpy as np

HERE = Path(__file__).resolve().parent
BUILD = HERE / "build"
CFLAGS = ["-O2", "-ffp-contract=off", "-fno-fast-math", "-fwrapv", "-fPIC", "-shared"]

_core = None
_fn_cache: dict[tuple, ctypes.CDLL] = {}


def build_core() -> Path:
    """Compile liboracle_core.so (idempotent)."""
    BUILD.mkdir(exist_ok=True)
    src = HERE / "oracle_core.c"
    out = BUILD / "liboracle_core.so"
    if not out.exists() or out.stat().st_mtime < src.stat().st_mtime:
        tmp = out.with_suffix(f".tmp{os.getpid()}")
        subprocess.run(["gcc", "-std=c11", *CFLAGS, str(src), "-o", str(tmp), "-lm"], check=True)
        os.replace(tmp, out)
    return out


def core() -> ctypes.CDLL:
    global _core
    if _core is None:
        lib = ctypes.CDLL(str(build_core()))
        P = ctypes.c_void_p
        lib.oracle_mandelbrot.argtypes = [P, P, ctypes.c_size_t, ctypes.c_int32]
        lib.oracle_compute_path.argtypes = [P, P, ctypes.c_int, ctypes.c_int, ctypes.c_int, P, P,
                                            ctypes.c_long]
        lib.oracle_compute_path.restype = ctypes.c_long
        lib.oracle_lmosem_error_image.argtypes = [P, ctypes.c_size_t, P, P, ctypes.c_int,
                                                  ctypes.c_int, ctypes.c_int]
        lib.oracle_lmosem_error_image.restype = ctypes.c_int64
        lib.oracle_lmosem_update.argtypes = [P, P, ctypes.c_size_t]
        lib.oracle_sum_f32_exact.argtypes = [P, ctypes.c_size_t]
        lib.oracle_sum_f32_exact.restype = ctypes.c_double
        lib.oracle_abssum_f32.argtypes = [P, ctypes.c_size_t]
        lib.oracle_abssum_f32.restype = ctypes.c_double
        lib.oracle_exscan_f32_exact.argtypes = [P, P, P, ctypes.c_size_t]
        lib.oracle_exscan_f32_seeded.argtypes = [P, P, ctypes.c_size_t, ctypes.c_double]
        lib.oracle_exscan_f32_sampled.argtypes = [P, ctypes.c_size_t, P, ctypes.c_size_t, P, P]
        _core = lib
    return _core


def _ptr(a: np.ndarray) -> int:
    assert a.flags["C_CONTIGUOUS"]
    return a.ctypes.data


# ---------------------------------------------------------------------------
# user functions (skeleton definitions, eqs. (1)-(4))
# ---------------------------------------------------------------------------
_PRELUDE = """
#define __global
#define __local
#define __constant
#define __private
#define __kernel
#include <math.h>
#include <stdint.h>
"""

_ENTRY = {
    "map": 'extern "C" void oracle_entry(const void* in, const void* in2, void* out, size_t n, '
           'const void* id, void** args) {{ (void)in2; (void)id; '
           'skel_oracle::map(&{f}, in, out, n, args); }}',
    "zip": 'extern "C" void oracle_entry(const void* in, const void* in2, void* out, size_t n, '
           'const void* id, void** args) {{ (void)id; '
           'skel_oracle::zip(&{f}, in, in2, out, n, args); }}',
    "reduce": 'extern "C" void oracle_entry(const void* in, const void* in2, void* out, size_t n, '
              'const void* id, void** args) {{ (void)in2; (void)id; '
              'skel_oracle::reduce(&{f}, in, out, n, args); }}',
    "scan": 'extern "C" void oracle_entry(const void* in, const void* in2, void* out, size_t n, '
            'const void* id, void** args) {{ (void)in2; '
            'skel_oracle::scan(&{f}, in, out, n, id, args); }}',
}
_SIZES = ('extern "C" void oracle_sizes(size_t* out, int* np) '
          '{{ skel_oracle::sizes_of(&{f}, out, np); }}')


def _strip_comments(src: str) -> str:
    src = re.sub(r"/\*.*?\*/", " ", src, flags=re.S)
    src = re.sub(r"//[^\n]*", " ", src)
    src = re.sub(r'"(\\.|[^"\\])*"', '""', src)
    return re.sub(r"^\s*#[^\n]*", " ", src, flags=re.M)


def entry_name(src: str) -> str:
    """The oracle is told nothing but the text: the user function is the last
    top-level function definition in it (the convention stated in DESIGN.md §1)."""
    src = _strip_comments(src)
    names = re.findall(r"([A-Za-z_]\w*)\s*\([^;{}]*\)\s*\{", src)
    names = [n for n in names if n not in ("if", "for", "while", "switch", "return")]
    if not names:
        raise ValueError("no function definition in user source")
    # the last definition at brace depth 0
    depth, last = 0, None
    pat = re.compile(r"([A-Za-z_]\w*)\s*\([^;{}]*\)\s*\{|\{|\}")
    for m in pat.finditer(src):
        tok = m.group(0)
        if m.group(1) is not None:
            if depth == 0 and m.group(1) not in ("if", "for", "while", "switch"):
                last = m.group(1)
            depth += 1
        elif tok == "{":
            depth += 1
        else:
            depth -= 1
    if last is None:
        raise ValueError("no top-level function definition in user source")
    return last


def _user_lib(src: str, kind: str, fname: str | None = None) -> ctypes.CDLL:
    fname = fname or entry_name(src)
    key = (src, kind, fname)
    if key in _fn_cache:
        return _fn_cache[key]
    BUILD.mkdir(exist_ok=True)
    text = "\n".join([_PRELUDE, src, f'#include "{HERE / "skel_oracle_impl.hpp"}"',
                      _ENTRY[kind].format(f=fname), _SIZES.format(f=fname), ""])
    h = hashlib.sha256(text.encode()).hexdigest()[:20]
    so = BUILD / f"uf_{kind}_{h}.so"
    if not so.exists():
        cpp = BUILD / f"uf_{kind}_{h}.cpp"
        cpp.write_text(text)
        tmp = so.with_suffix(f".tmp{os.getpid()}")
        r = subprocess.run(["g++", "-std=c++17", *CFLAGS, str(cpp), "-o", str(tmp)],
                           capture_output=True, text=True)
        if r.returncode != 0:
            raise SyntaxError(f"oracle: user function does not compile:\n{r.stderr}")
        os.replace(tmp, so)
    lib = ctypes.CDLL(str(so))
    P = ctypes.c_void_p
    lib.oracle_entry.argtypes = [P, P, P, ctypes.c_size_t, P, P]
    lib.oracle_sizes.argtypes = [P, P]
    _fn_cache[key] = lib
    return lib


def _sizes(lib) -> tuple[int, list[int]]:
    buf = (ctypes.c_size_t * 64)()
    npar = ctypes.c_int()
    lib.oracle_sizes(buf, ctypes.byref(npar))
    return int(buf[0]), [int(buf[i + 1]) for i in range(npar.value)]


def _pack_args(args, expect: list[int]):
    """Arguments object: vectors by pointer, everything else by bytes."""
    keep = []
    arr = (ctypes.c_void_p * max(1, len(args)))()
    if len(args) != len(expect):
        raise TypeError(f"user function takes {len(expect)} extra arguments, got {len(args)}")
    for i, (a, sz) in enumerate(zip(args, expect)):
        if isinstance(a, np.ndarray) and a.ndim >= 1:
            if sz != 0:
                raise TypeError(f"argument {i}: vector passed for a by-value parameter")
            arr[i] = _ptr(a)
        else:
            b = np.asarray(a)
            if b.dtype.itemsize != sz:
                raise TypeError(f"argument {i}: {b.dtype.itemsize} bytes, parameter has {sz}")
            b = np.ascontiguousarray(b.reshape(1))
            keep.append(b)
            arr[i] = _ptr(b)
    return arr, keep


def skel_map(src: str, x: np.ndarray, out_dtype=None, args=(), fname=None):
    """eq. (1): [f(x_0), ..., f(x_{n-1})]; void f -> returns None (side effects)."""
    lib = _user_lib(src, "map", fname)
    rsz, psz = _sizes(lib)
    if psz[0] != x.dtype.itemsize:
        raise TypeError("element size mismatch")
    argv, keep = _pack_args(list(args), psz[1:])
    x = np.ascontiguousarray(x)
    if rsz == 0:
        lib.oracle_entry(_ptr(x), None, None, x.size, None, argv)
        return None
    out = np.empty(x.size, dtype=out_dtype)
    assert out.dtype.itemsize == rsz
    lib.oracle_entry(_ptr(x), None, _ptr(out), x.size, None, argv)
    return out


def skel_zip(src: str, a: np.ndarray, b: np.ndarray, out_dtype, args=(), fname=None):
    """eq. (2): [x_0 (+) y_0, ..., x_{n-1} (+) y_{n-1}] for equally sized inputs."""
    if a.size != b.size:
        raise ValueError("zip: vectors must have equal sizes (P:L268-269)")
    lib = _user_lib(src, "zip", fname)
    rsz, psz = _sizes(lib)
    argv, keep = _pack_args(list(args), psz[2:])
    a = np.ascontiguousarray(a)
    b = np.ascontiguousarray(b)
    out = np.empty(a.size, dtype=out_dtype)
    assert out.dtype.itemsize == rsz
    lib.oracle_entry(_ptr(a), _ptr(b), _ptr(out), a.size, None, argv)
    return out


def skel_reduce(src: str, x: np.ndarray, args=(), fname=None):
    """eq. (3) as the left fold x_0 (+) x_1 (+) ... (+) x_{n-1}; n = 0 is an error."""
    if x.size == 0:
        raise ValueError("reduce of an empty vector is undefined (eq. 3 has no identity)")
    lib = _user_lib(src, "reduce", fname)
    rsz, psz = _sizes(lib)
    argv, keep = _pack_args(list(args), psz[2:])
    x = np.ascontiguousarray(x)
    out = np.empty(1, dtype=x.dtype)
    lib.oracle_entry(_ptr(x), None, _ptr(out), x.size, None, argv)
    return out[0]


def skel_scan(src: str, x: np.ndarray, identity, args=(), fname=None):
    """eq. (4): [id, x_0, x_0(+)x_1, ..., x_0(+)...(+)x_{n-2}] (exclusive)."""
    lib = _user_lib(src, "scan", fname)
    rsz, psz = _sizes(lib)
    argv, keep = _pack_args(list(args), psz[2:])
    x = np.ascontiguousarray(x)
    out = np.empty(x.size, dtype=x.dtype)
    idv = np.ascontiguousarray(np.asarray(identity, dtype=x.dtype).reshape(1))
    if x.size:
        lib.oracle_entry(_ptr(x), None, _ptr(out), x.size, _ptr(idv), argv)
    return out


# ---------------------------------------------------------------------------
# float '+' Reduce / Scan reference values (reading R2)
# ---------------------------------------------------------------------------
def sum_f32_exact(x: np.ndarray) -> float:
    x = np.ascontiguousarray(x, dtype=np.float32)
    return core().oracle_sum_f32_exact(_ptr(x), x.size)


def abssum_f32(x: np.ndarray) -> float:
    x = np.ascontiguousarray(x, dtype=np.float32)
    return core().oracle_abssum_f32(_ptr(x), x.size)


def exscan_f32_exact(x: np.ndarray):
    """Returns (prefix sums rounded to float32, sum_{j<i} |x_j| in float64)."""
    x = np.ascontiguousarray(x, dtype=np.float32)
    out = np.empty(x.size, np.float32)
    ab = np.empty(x.size, np.float64)
    if x.size:
        core().oracle_exscan_f32_exact(_ptr(x), _ptr(out), _ptr(ab), x.size)
    return out, ab


def exscan_f32_seeded(x: np.ndarray, s0: float, out: np.ndarray | None = None) -> np.ndarray:
    """Exclusive float '+' scan of a chunk whose preceding elements sum to s0."""
    x = np.ascontiguousarray(x, dtype=np.float32)
    if out is None:
        out = np.empty(x.size, np.float32)
    if x.size:
        core().oracle_exscan_f32_seeded(_ptr(x), _ptr(out), x.size, float(s0))
    return out


def exscan_f32_sampled(x: np.ndarray, idx: np.ndarray):
    """Exact (float64) exclusive prefix sums of x at the sorted positions idx."""
    x = np.ascontiguousarray(x, dtype=np.float32)
    idx = np.ascontiguousarray(np.sort(idx), dtype=np.int64)
    pre = np.empty(idx.size, np.float64)
    ab = np.empty(idx.size, np.float64)
    core().oracle_exscan_f32_sampled(_ptr(x), x.size, _ptr(idx), idx.size, _ptr(pre), _ptr(ab))
    return idx, pre, ab


# ---------------------------------------------------------------------------
# workloads
# ---------------------------------------------------------------------------
def mandelbrot(pos: np.ndarray, cap: int) -> np.ndarray:
    """eq. (5) escape-time counts for a Vector<{float re, im}> of positions."""
    pos = np.ascontiguousarray(pos)
    assert pos.dtype.itemsize == 8
    out = np.empty(pos.size, np.int32)
    core().oracle_mandelbrot(_ptr(pos), _ptr(out), pos.size, cap)
    return out


def compute_path(p1, p2, dims=(150, 150, 280)):
    """Siddon merged-alpha path: (coords int64[], lens float64[])."""
    a = np.ascontiguousarray(p1, dtype=np.float64)
    b = np.ascontiguousarray(p2, dtype=np.float64)
    cap = sum(dims) + 3
    coord = np.empty(cap, np.int64)
    ln = np.empty(cap, np.float64)
    m = core().oracle_compute_path(_ptr(a), _ptr(b), *dims, _ptr(coord), _ptr(ln), cap)
    assert m >= 0
    return coord[:m].copy(), ln[:m].copy()


def lmosem_error_image(events: np.ndarray, f: np.ndarray, dims=(150, 150, 280), c=None):
    """Listing 3 lines 4-13 for one subset; returns (c float64, n_valid)."""
    ev = np.ascontiguousarray(events)
    assert ev.dtype.itemsize == 24
    f64 = np.ascontiguousarray(f, dtype=np.float64)
    if c is None:
        c = np.zeros(int(np.prod(dims)), np.float64)
    nv = core().oracle_lmosem_error_image(_ptr(ev), ev.size, _ptr(f64), _ptr(c), *dims)
    return c, int(nv)


def lmosem_update(f: np.ndarray, c: np.ndarray) -> np.ndarray:
    """Listing 3 lines 14-16: f[j] *= c[j] where c[j] > 0 (returns a new array)."""
    f = np.array(f, dtype=np.float64, copy=True)
    c = np.ascontiguousarray(c, dtype=np.float64)
    core().oracle_lmosem_update(_ptr(f), _ptr(c), f.size)
    return f


def lmosem_subset(events: np.ndarray, f: np.ndarray, dims=(150, 150, 280)):
    """One subset iteration of Listing 3 with c reset to 0 (reading R10(i))."""
    c, nv = lmosem_error_image(events, f, dims)
    return lmosem_update(f, c), c, nv


def lmosem_reconstruct(subsets, dims=(150, 150, 280), f0=1.0):
    """Listing 3's outer loop over the subsets; f0 = 1 everywhere (reading R10(ii))."""
    f = np.full(int(np.prod(dims)), f0, np.float64)
    for ev in subsets:
        f, _, _ = lmosem_subset(ev, f, dims)
    return f
