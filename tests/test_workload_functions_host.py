"""The LM OSEM customizing function (workloads/lmosem_error.cu) is plain C++
apart from atomicAdd/__ldg/float4; compiled for the host with a few one-line shims
it can be checked against the oracle on the CPU (tiny grids with exact
plane/edge/corner ties, and the paper-sized volume).  This tests the walk's
logic only; the GPU parity tests run the same text through NVRTC."""
import ctypes
import subprocess
from pathlib import Path

import numpy as np
import pytest

import oracle
import skel_inputs as si

ROOT = Path(__file__).resolve().parents[1]
SHIM = r'''
#include <cmath>
#include <algorithm>
using std::min; using std::max; using std::fmin; using std::fmax;
#define __forceinline__ inline
template <class T> static T __ldg(const T* p) { return *p; }
struct float4 { float x, y, z, w; };
static inline float4 make_float4(float a, float b, float c, float d) { return float4{a, b, c, d}; }
#include "SRC"
extern "C" void run(const float* ev, int n, const float* f, float* c, int nx, int ny, int nz) {
    for (int i = 0; i < n; ++i) {
        Event e{ev[6*i], ev[6*i+1], ev[6*i+2], ev[6*i+3], ev[6*i+4], ev[6*i+5]};
        lmosem_error(e, f, c, nx, ny, nz);
    }
}
// the lanes form (workloads/lmosem_lanes.cu) with the group sum done in lane order
extern "C" void run_lanes(const float* ev, int n, const float* f, float* c, int nx, int ny, int nz, int lanes) {
    for (int i = 0; i < n; ++i) {
        Event e{ev[6*i], ev[6*i+1], ev[6*i+2], ev[6*i+3], ev[6*i+4], ev[6*i+5]};
        Walk w[32];
        bool ok[32];
        float fp = 0.0f;
        for (int l = 0; l < lanes; ++l) {
            ok[l] = walk_piece(e, nx, ny, nz, l, lanes, w[l]);
            if (ok[l]) fp += forward(w[l], f);
        }
        if (!(fp > 0.0f)) continue;
        for (int l = 0; l < lanes; ++l)
            if (ok[l]) back_project(w[l], c, 1.0f / fp);
    }
}
'''


@pytest.fixture(scope="module")
def walk(tmp_path_factory):
    d = tmp_path_factory.mktemp("walk")
    src = d / "shim.cpp"
    src.write_text(SHIM.replace("SRC", str(ROOT / "paper_conf_ipps_steuwerkg11_b200" / "workloads" / "lmosem_error.cu")))
    so = d / "walk.so"
    subprocess.run(["g++", "-O2", "-std=c++17", "-ffp-contract=off", "-shared", "-fPIC", str(src), "-o", str(so)],
                   check=True)
    lib = ctypes.CDLL(str(so))
    P, I = ctypes.c_void_p, ctypes.c_int
    lib.run.argtypes = [P, I, P, P, I, I, I]
    lib.run_lanes.argtypes = [P, I, P, P, I, I, I, I]

    def run(ev, f, dims, lanes=0):
        c = np.zeros(int(np.prod(dims)), np.float32)
        f32 = np.ascontiguousarray(f, np.float32)
        if lanes:
            lib.run_lanes(ev.ctypes.data, ev.size, f32.ctypes.data, c.ctypes.data, *dims, lanes)
        else:
            lib.run(ev.ctypes.data, ev.size, f32.ctypes.data, c.ctypes.data, *dims)
        return c
    return run


@pytest.mark.parametrize("quarter", [False, True])
def test_tiny_grid_with_ties(walk, quarter):
    g = np.random.default_rng(5 + quarter)
    dims = (4, 3, 5)
    e = np.zeros(500, si.EVENT_DTYPE)
    for k in ("x1", "y1", "z1", "x2", "y2", "z2"):
        e[k] = g.integers(-8, 28, 500) / 4.0 if quarter else g.uniform(-2, 7, 500)
    f = g.uniform(0.5, 2, int(np.prod(dims))).astype(np.float32)
    c = walk(e, f, dims)
    want, _ = oracle.lmosem_error_image(e, f.astype(np.float64), dims)
    assert np.array_equal(c > 0, want > 0)  # same voxels touched
    assert np.linalg.norm(c - want) <= 1e-6 * np.linalg.norm(want)


@pytest.mark.parametrize("lanes", [2, 3, 4, 8, 32])
@pytest.mark.parametrize("quarter", [False, True])
def test_lanes_pieces_tiny_grid_with_ties(walk, quarter, lanes):
    """lmosem_lanes: `lanes` alpha pieces per line of response, partial forward
    projections summed, each piece back-projected -- the same error image as
    the oracle (Listing 3) on grids with exact plane/edge/corner ties
    (quarter-voxel endpoints put piece boundaries on planes too)."""
    g = np.random.default_rng(15 + quarter)
    dims = (4, 3, 5)
    e = np.zeros(500, si.EVENT_DTYPE)
    for k in ("x1", "y1", "z1", "x2", "y2", "z2"):
        e[k] = g.integers(-8, 28, 500) / 4.0 if quarter else g.uniform(-2, 7, 500)
    f = g.uniform(0.5, 2, int(np.prod(dims))).astype(np.float32)
    c = walk(e, f, dims, lanes=lanes)
    want, _ = oracle.lmosem_error_image(e, f.astype(np.float64), dims)
    assert np.array_equal(c > 0, want > 0)
    # up to 32 float32 partial sums per fp and two reductions per cut voxel:
    # a few float32 roundings more than the one-walk form (1e-6)
    assert np.linalg.norm(c - want) <= 1e-5 * np.linalg.norm(want)


@pytest.mark.parametrize("lanes", [4, 8])
def test_lanes_pieces_paper_volume(walk, lanes):
    ev = si.lmosem_events(5000, subset=5)
    dims = (150, 150, 280)
    c = walk(ev, np.ones(int(np.prod(dims))), dims, lanes=lanes)
    want, _ = oracle.lmosem_error_image(ev, np.ones(int(np.prod(dims))), dims)
    assert np.array_equal(c > 0, want > 0)
    assert np.linalg.norm(c - want) <= 1e-6 * np.linalg.norm(want)


def test_paper_volume_no_flips(walk):
    ev = si.lmosem_events(5000, subset=4)
    dims = (150, 150, 280)
    c = walk(ev, np.ones(int(np.prod(dims))), dims)
    want, _ = oracle.lmosem_error_image(ev, np.ones(int(np.prod(dims))), dims)
    assert np.array_equal(c > 0, want > 0)
    assert np.linalg.norm(c - want) <= 1e-6 * np.linalg.norm(want)


MANDEL_SHIM = r'''
#include "SRC"
extern "C" void run(const float* pos, long n, int cap, int* out) {
    for (long i = 0; i < n; ++i) out[i] = mandelbrot_blocked(Pos{pos[2*i], pos[2*i+1]}, cap);
}
'''


@pytest.fixture(scope="module")
def mandel_blocked(tmp_path_factory):
    d = tmp_path_factory.mktemp("mandel")
    src = d / "shim.cpp"
    src.write_text(MANDEL_SHIM.replace(
        "SRC", str(ROOT / "paper_conf_ipps_steuwerkg11_b200" / "workloads" / "mandelbrot_blocked.cu")))
    so = d / "mandel.so"
    subprocess.run(["g++", "-O2", "-std=c++17", "-ffp-contract=off", "-shared", "-fPIC", str(src), "-o", str(so)],
                   check=True)
    lib = ctypes.CDLL(str(so))
    lib.run.argtypes = [ctypes.c_void_p, ctypes.c_long, ctypes.c_int, ctypes.c_void_p]

    def run(pos, cap):
        pos = np.ascontiguousarray(pos)
        out = np.zeros(pos.size, np.int32)
        lib.run(pos.ctypes.data, pos.size, cap, out.ctypes.data)
        return out
    return run


BLOCKED_FORMS = {
    "periodic": "#define MANDEL_PERIODIC 1\n#define MANDEL_PRE 8\n",
    "maxtest": "#define MANDEL_MAXTEST 1\n",
    "fsetp": "#define MANDEL_MAXTEST 0\n",
    "fsetp_periodic": "#define MANDEL_MAXTEST 0\n#define MANDEL_PERIODIC 1\n#define MANDEL_PRE 8\n",
    "maxtest_periodic": "#define MANDEL_MAXTEST 1\n#define MANDEL_PERIODIC 1\n#define MANDEL_PRE 8\n",
    "maxtest_blockstart": "#define MANDEL_MAXTEST 1\n#define MANDEL_PERIODIC 2\n#define MANDEL_PRE 8\n",
    "maxtest_blockstart_b4": "#define MANDEL_MAXTEST 1\n#define MANDEL_PERIODIC 2\n#define MANDEL_B 4\n",
    "noreplay": "#define MANDEL_NOREPLAY 1\n",
    "noreplay_periodic": "#define MANDEL_NOREPLAY 1\n#define MANDEL_PERIODIC 1\n",
    "noreplay_periodic_b4": "#define MANDEL_NOREPLAY 1\n#define MANDEL_PERIODIC 1\n#define MANDEL_B 4\n",
}


@pytest.mark.parametrize("form", sorted(BLOCKED_FORMS))
@pytest.mark.parametrize("cap", [1, 7, 8, 9, 17, 256, 1024, 1500])
def test_blocked_forms_equal_the_plain_iteration(tmp_path, golden_dir, cap, form):
    """mandelbrot_blocked.cu in its other forms -- exact periodicity checking
    (Brent's save schedule at block ends) with an 8-update plain prefix, the
    block's tests folded into one NaN-propagating maximum (MANDEL_MAXTEST), and
    blocks that keep their test values so an escape needs no replay
    (MANDEL_NOREPLAY): the counts of eq. (5) as written on the whole 1024x768
    image, and the golden CRC at cap 256."""
    import json
    import os
    import zlib
    src = tmp_path / "periodic.cpp"
    src.write_text(BLOCKED_FORMS[form] + MANDEL_SHIM.replace(
        "SRC", str(ROOT / "paper_conf_ipps_steuwerkg11_b200" / "workloads" / "mandelbrot_blocked.cu")))
    so = tmp_path / "periodic.so"
    subprocess.run(["g++", "-O2", "-std=c++17", "-ffp-contract=off", "-shared", "-fPIC", str(src), "-o", str(so)],
                   check=True)
    lib = ctypes.CDLL(str(so))
    lib.run.argtypes = [ctypes.c_void_p, ctypes.c_long, ctypes.c_int, ctypes.c_void_p]
    pos = np.ascontiguousarray(si.mandelbrot_positions(1024, 768))
    got = np.zeros(pos.size, np.int32)
    lib.run(pos.ctypes.data, pos.size, cap, got.ctypes.data)
    assert np.array_equal(got, oracle.mandelbrot(pos, cap))
    if cap == 256:
        with open(os.path.join(golden_dir, "mandelbrot.json")) as fh:
            case = [c for c in json.load(fh)["cases"] if (c["width"], c["height"], c["cap"]) == (1024, 768, 256)][0]
        assert zlib.crc32(got.tobytes()) == int(case["crc32"], 16)


@pytest.mark.parametrize("cap", [1, 7, 8, 9, 256, 1024, 1500])
def test_blocked_mandelbrot_equals_the_plain_iteration(mandel_blocked, golden_dir, cap):
    """mandelbrot_blocked.cu (loop control per block of 8 updates, roll back on
    escape) counts exactly what eq. (5) as written counts: bit-identical to
    the oracle on the whole 1024x768 image, for caps below, at and above the
    block size, and to the golden CRC at cap 256."""
    import json
    import os
    import zlib
    pos = si.mandelbrot_positions(1024, 768)
    got = mandel_blocked(pos, cap)
    assert np.array_equal(got, oracle.mandelbrot(pos, cap))
    if cap == 256:
        with open(os.path.join(golden_dir, "mandelbrot.json")) as fh:
            case = [c for c in json.load(fh)["cases"] if (c["width"], c["height"], c["cap"]) == (1024, 768, 256)][0]
        assert zlib.crc32(got.tobytes()) == int(case["crc32"], 16)


ORDER_SHIM = r'''
#include <cmath>
#include <algorithm>
using std::min; using std::max; using std::fmin; using std::fmax; using std::fabs;
#define __forceinline__ inline
template <class T> static T __ldg(const T* p) { return *p; }
struct float4 { float x, y, z, w; };
static inline float4 make_float4(float a, float b, float c, float d) { return float4{a, b, c, d}; }
#include <cstring>
static inline unsigned __float_as_uint(float f) { unsigned u; std::memcpy(&u, &f, 4); return u; }
#include "ERR"
#include "ORD"
extern "C" void buckets(const float* ev, int n, int nx, int ny, int nz, int nb, int* out) {
    for (int i = 0; i < n; ++i) {
        Event e{ev[6*i], ev[6*i+1], ev[6*i+2], ev[6*i+3], ev[6*i+4], ev[6*i+5]};
        out[i] = lm_bucket(e, nx, ny, nz, nb);
    }
}
'''


def test_device_order_key_follows_the_exact_path_length(tmp_path):
    """lm_bucket (workloads/lmosem_order.cu, the key of the on-device event
    ordering): bucket 0 = longest clipped path; checked against the oracle's
    exact Siddon path lengths (rank correlation), range [0, nb), and a ray that
    misses the volume goes last."""
    wl = ROOT / "paper_conf_ipps_steuwerkg11_b200" / "workloads"
    src = tmp_path / "order.cpp"
    src.write_text(ORDER_SHIM.replace("ERR", str(wl / "lmosem_error.cu")).replace("ORD", str(wl / "lmosem_order.cu")))
    so = tmp_path / "order.so"
    subprocess.run(["g++", "-O2", "-std=c++17", "-ffp-contract=off", "-shared", "-fPIC", str(src), "-o", str(so)],
                   check=True)
    lib = ctypes.CDLL(str(so))
    lib.buckets.argtypes = [ctypes.c_void_p, ctypes.c_int, ctypes.c_int, ctypes.c_int, ctypes.c_int, ctypes.c_int,
                            ctypes.c_void_p]
    ev = si.lmosem_events(3000, subset=5)
    miss = np.zeros(1, si.EVENT_DTYPE)
    miss["x1"], miss["y1"], miss["z1"], miss["x2"], miss["y2"], miss["z2"] = -5, -5, -5, -9, -1, -7
    ev = np.concatenate([ev, miss])
    nb = 64
    b = np.zeros(ev.size, np.int32)
    lib.buckets(ev.ctypes.data, ev.size, 150, 150, 280, nb, b.ctypes.data)
    assert b.min() >= 0 and b.max() <= nb - 1 and b[-1] == nb - 1
    # the walk's work is its voxel count: the oracle's number of path segments
    nvox = np.array([len(oracle.compute_path((e["x1"], e["y1"], e["z1"]), (e["x2"], e["y2"], e["z2"]))[0])
                     for e in ev[:-1]])
    from scipy.stats import spearmanr
    r = spearmanr(b[:-1], -nvox).statistic  # ties (a bucket holds many events) ranked by their mean
    assert r > 0.95, r


PAIRS_SHIM = r'''
#define __forceinline__ inline
#include "SRC"
extern "C" void run(const float* pos, long npairs, int cap, int* out) {
    for (long i = 0; i < npairs; ++i) {
        Cnt2 r = mandelbrot_pairs(Pos2{pos[4*i], pos[4*i+1], pos[4*i+2], pos[4*i+3]}, cap);
        out[2*i] = r.n0;
        out[2*i+1] = r.n1;
    }
}
'''


@pytest.mark.parametrize("maxtest", [False, True, "noreplay", "noreplay_fsetp"])
@pytest.mark.parametrize("periodic", [False, True])
@pytest.mark.parametrize("cap", [1, 5, 8, 9, 17, 256, 1500])
def test_pairs_mandelbrot_equals_the_plain_iteration(tmp_path, golden_dir, cap, periodic, maxtest):
    """mandelbrot_pairs.cu (two neighbouring pixels per element, packed updates
    emulated one float at a time on the host): bit-identical to eq. (5) as
    written (the oracle) on the whole 1024x768 image, caps below/at/above the
    prefix and block lengths, and to the golden CRC at cap 256."""
    import json
    import os
    import zlib
    src = tmp_path / "pairs.cpp"
    src.write_text(("#define MANDEL_PERIODIC 1\n" if periodic else "") +
                   ("#define MANDEL_MAXTEST 1\n" if maxtest else "#define MANDEL_MAXTEST 0\n") +
                   ("#define MANDEL_NOREPLAY 1\n" if str(maxtest).startswith("noreplay") else "") +
                   ("#define MANDEL_NR_FSETP 1\n" if maxtest == "noreplay_fsetp" else "") + PAIRS_SHIM.replace(
        "SRC", str(ROOT / "paper_conf_ipps_steuwerkg11_b200" / "workloads" / "mandelbrot_pairs.cu")))
    so = tmp_path / "pairs.so"
    subprocess.run(["g++", "-O2", "-std=c++17", "-ffp-contract=off", "-shared", "-fPIC", str(src), "-o", str(so)],
                   check=True)
    lib = ctypes.CDLL(str(so))
    lib.run.argtypes = [ctypes.c_void_p, ctypes.c_long, ctypes.c_int, ctypes.c_void_p]
    pos = np.ascontiguousarray(si.mandelbrot_positions(1024, 768))
    got = np.zeros(pos.size, np.int32)
    lib.run(pos.ctypes.data, pos.size // 2, cap, got.ctypes.data)
    assert np.array_equal(got, oracle.mandelbrot(pos, cap))
    if cap == 256:
        with open(os.path.join(golden_dir, "mandelbrot.json")) as fh:
            case = [c for c in json.load(fh)["cases"] if (c["width"], c["height"], c["cap"]) == (1024, 768, 256)][0]
        assert zlib.crc32(got.tobytes()) == int(case["crc32"], 16)
