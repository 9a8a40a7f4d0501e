"""GPU parity of the four skeletons (eqs. (1)-(4)) against the CPU oracle.

Bars (BASELINE.json north_star): bit-exact for integer data and
for float Map/Zip built from + - * / (FMA contraction off on both sides);
float Reduce/Scan within 1e-5 normwise: |gpu - exact| <= 1e-5 * sum |x|.
Sizes span several 64 KB tiles and ragged tails.
"""
import numpy as np
import pytest

import oracle
import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import (MAP_F32, MAP_I32, MULT_F32, SAXPY_F32, SAXPY_I32,
                                                         SUM_F32, SUM_I32)

pytestmark = pytest.mark.gpu

SIZES = [1, 3, 4, 5, 127, 4097, 16384, 16385, 3 * 16384 + 17, (1 << 20) + 3]

MAT_U = """
struct M2 { unsigned a, b, c, d; };   /* row-major 2x2 matrix, mod 2^32 */
M2 matmul(M2 x, M2 y) {
  M2 r;
  r.a = x.a*y.a + x.b*y.c;  r.b = x.a*y.b + x.b*y.d;
  r.c = x.c*y.a + x.d*y.c;  r.d = x.c*y.b + x.d*y.d;
  return r;
}
"""
M2 = np.dtype([("a", np.uint32), ("b", np.uint32), ("c", np.uint32), ("d", np.uint32)])
# 12-byte element (not a TMA-friendly size): affine maps x -> a*x + b composed
# left to right, plus a count -- associative, not commutative
AFF3 = """
struct Aff { unsigned a, b, n; };
Aff compose(Aff f, Aff g) { Aff r; r.a = f.a * g.a; r.b = f.b * g.a + g.b; r.n = f.n + g.n; return r; }
"""
AFF = np.dtype([("a", np.uint32), ("b", np.uint32), ("n", np.uint32)])
# 8-byte element: affine composition in uint32 pairs
AFF2 = """
struct A2 { unsigned a, b; };
A2 comp2(A2 f, A2 g) { A2 r; r.a = f.a * g.a; r.b = f.b * g.a + g.b; return r; }
"""
A2 = np.dtype([("a", np.uint32), ("b", np.uint32)])


@pytest.fixture(scope="module")
def ctx():
    c = skel.Context(1)
    yield c
    c.close()


def rand_struct(dt, n, seed):
    g = np.random.default_rng(seed)
    out = np.zeros(n, dt)
    for k in dt.names:
        out[k] = g.integers(0, 1 << 32, n, dtype=np.uint64).astype(np.uint32)
    return out


# ---- Map / Zip ----------------------------------------------------------------
@pytest.mark.parametrize("n", SIZES)
def test_map_f32_bit_exact(ctx, n):
    x = si.uniform_f32(n, 20110516 + n % 97)
    out = ctx.vector(n=n, dtype=np.float32)
    ctx.map(MAP_F32, ctx.vector(x), out)
    assert np.array_equal(out.download(), oracle.skel_map(MAP_F32, x, np.float32))


@pytest.mark.parametrize("n", [1, 5, 4097, (1 << 20) + 3])
def test_map_i32_bit_exact(ctx, n):
    x = si.uniform_i32(n, 7)
    out = ctx.vector(n=n, dtype=np.int32)
    ctx.map(MAP_I32, ctx.vector(x), out)
    assert np.array_equal(out.download(), oracle.skel_map(MAP_I32, x, np.int32))


@pytest.mark.parametrize("n", SIZES)
def test_zip_saxpy_f32_bit_exact(ctx, n):
    x, y = si.uniform_f32(n, 1), si.uniform_f32(n, 2)
    out = ctx.vector(n=n, dtype=np.float32)
    ctx.zip(SAXPY_F32, ctx.vector(x), ctx.vector(y), out, args=[np.float32(2.5)])
    want = oracle.skel_zip(SAXPY_F32, x, y, np.float32, args=[np.float32(2.5)])
    assert np.array_equal(out.download(), want)


@pytest.mark.parametrize("n", [3, 4097, (1 << 20) + 3])
def test_zip_saxpy_i32_bit_exact(ctx, n):
    x, y = si.uniform_i32(n, 3), si.uniform_i32(n, 4)
    out = ctx.vector(n=n, dtype=np.int32)
    ctx.zip(SAXPY_I32, ctx.vector(x), ctx.vector(y), out, args=[np.int32(3)])
    want = oracle.skel_zip(SAXPY_I32, x, y, np.int32, args=[np.int32(3)])
    assert np.array_equal(out.download(), want)


def test_map_struct_element_and_helpers(ctx):
    src = """
    struct Pos { float re, im; };
    float sq(float v) { return v * v; }
    float norm2(Pos p) { return sq(p.re) + sq(p.im); }
    """
    pos = si.mandelbrot_positions(64, 48)
    out = ctx.vector(n=pos.size, dtype=np.float32)
    ctx.map(src, ctx.vector(pos), out)
    assert np.array_equal(out.download(), oracle.skel_map(src, pos, np.float32))


def test_map_listing2_argument(ctx):
    src = "float f(float input, float number) { return input * number; }"
    x = si.uniform_f32(1000, 5)
    out = ctx.vector(n=x.size, dtype=np.float32)
    ctx.map(src, ctx.vector(x), out, args=[np.float32(5)])
    assert np.array_equal(out.download(), oracle.skel_map(src, x, np.float32, args=[np.float32(5)]))


def test_argument_order_and_mixed_kinds(ctx):
    src = """
    float g(float x, double a, int k, const float* tab, float b) { return (float)(a * x) - b * tab[k]; }
    """
    x = si.uniform_f32(5000, 9)
    tab = np.arange(8, dtype=np.float32) + 1
    args_gpu = [np.float64(3.0), np.int32(5), ctx.vector(tab), np.float32(0.5)]
    args_cpu = [np.float64(3.0), np.int32(5), tab, np.float32(0.5)]
    out = ctx.vector(n=x.size, dtype=np.float32)
    ctx.map(src, ctx.vector(x), out, args=args_gpu)
    assert np.array_equal(out.download(), oracle.skel_map(src, x, np.float32, args=args_cpu))


def test_void_map_side_effect(ctx):
    src = "void h(int x, int* hist) { atomicAdd(&hist[x], 1); }"
    x = np.random.default_rng(0).integers(0, 16, 100_000).astype(np.int32)
    hist = ctx.vector(n=16, dtype=np.int32)
    ctx.map(src, ctx.vector(x), None, args=[hist])
    hist.mark_device_modified()
    assert np.array_equal(hist.download(), np.bincount(x, minlength=16).astype(np.int32))


def test_inplace_map(ctx):
    x = si.uniform_f32(70_001, 3)
    v = ctx.vector(x)
    ctx.map(MAP_F32, v, v)
    assert np.array_equal(v.download(), oracle.skel_map(MAP_F32, x, np.float32))


def test_empty_vectors(ctx):
    v = ctx.vector(n=0, dtype=np.float32)
    o = ctx.vector(n=0, dtype=np.float32)
    ctx.map(MAP_F32, v, o)
    ctx.scan(SUM_F32, v, o, np.float32(0))
    assert o.download().size == 0
    with pytest.raises(skel.SkelError) as e:
        ctx.reduce(SUM_F32, v)
    assert e.value.name == "SKEL_ERR_SIZE"


def test_error_paths(ctx):
    a = ctx.vector(np.ones(3, np.float32))
    b = ctx.vector(np.ones(4, np.float32))
    with pytest.raises(skel.SkelError) as e:
        ctx.zip(MULT_F32, a, b, ctx.vector(n=3, dtype=np.float32))
    assert e.value.name == "SKEL_ERR_SIZE"
    with pytest.raises(skel.SkelError) as e:  # Listing 2 as printed (missing ';')
        ctx.map("float f(float input, float number) { return input * number }", a,
                ctx.vector(n=3, dtype=np.float32), args=[np.float32(5)])
    assert e.value.name == "SKEL_ERR_COMPILE" and 'expected a ";"' in e.value.msg
    with pytest.raises(skel.SkelError) as e:  # double vector into a float function
        ctx.map(MAP_F32, ctx.vector(np.ones(3, np.float64)), ctx.vector(n=3, dtype=np.float32))
    assert e.value.name == "SKEL_ERR_TYPE"
    with pytest.raises(skel.SkelError) as e:  # missing argument
        ctx.zip(SAXPY_F32, a, a, ctx.vector(n=3, dtype=np.float32))
    assert e.value.name == "SKEL_ERR_TYPE"
    with pytest.raises(skel.SkelError) as e:  # scalar of the wrong size
        ctx.zip(SAXPY_F32, a, a, ctx.vector(n=3, dtype=np.float32), args=[np.float64(1)])
    assert e.value.name == "SKEL_ERR_TYPE"


# ---- Reduce ---------------------------------------------------------------------
def assert_sum_close(got, x):
    exact = oracle.sum_f32_exact(x)
    scale = oracle.abssum_f32(x)
    assert abs(float(got) - exact) <= 1e-5 * scale + 1e-30, (float(got), exact)


@pytest.mark.parametrize("n", SIZES)
def test_reduce_sum_f32(ctx, n):
    x = si.uniform_f32(n, 11 + n % 13)
    assert_sum_close(ctx.reduce(SUM_F32, ctx.vector(x)), x)


# signed data and cancellation: the normwise bar's scale is
# sum |x_i|; U[0,1) data alone would not notice a dropped |.| anywhere
SIGNED_SIZES = [1, 5, 16385, (1 << 20) + 3, (1 << 26) + 3]


@pytest.mark.parametrize("n", SIGNED_SIZES)
@pytest.mark.parametrize("gen", ["signed", "cancel"])
def test_reduce_sum_f32_signed(ctx, n, gen):
    x = (si.uniform_signed_f32 if gen == "signed" else si.cancellation_f32)(n, 40 + n % 11)
    assert_sum_close(ctx.reduce(SUM_F32, ctx.vector(x)), x)


@pytest.mark.parametrize("n", SIZES)
def test_reduce_sum_i32_exact(ctx, n):
    x = si.uniform_int01(n, 5)
    assert int(ctx.reduce(SUM_I32, ctx.vector(x))) == int(oracle.skel_reduce(SUM_I32, x))


def test_reduce_arange_closed_form(ctx):
    n = 5793  # every partial sum < 2^24: any association order is exact
    assert float(ctx.reduce(SUM_F32, ctx.vector(np.arange(n, dtype=np.float32)))) == n * (n - 1) // 2


@pytest.mark.parametrize("n", [1, 2, 33, 4097, 8192, 8193, 5 * 8192 + 3, 300_001])
def test_reduce_noncommutative_16B(ctx, n):
    m = rand_struct(M2, n, n)
    got = ctx.reduce(MAT_U, ctx.vector(m))
    want = oracle.skel_reduce(MAT_U, m)
    assert got.tobytes() == want.tobytes()


@pytest.mark.parametrize("n", [1, 7, 16384, 16385, 200_003])
def test_reduce_noncommutative_8B(ctx, n):
    m = rand_struct(A2, n, n + 1)
    assert ctx.reduce(AFF2, ctx.vector(m)).tobytes() == oracle.skel_reduce(AFF2, m).tobytes()


@pytest.mark.parametrize("n", [1, 9, 5461, 5462, 100_001])
def test_reduce_noncommutative_12B_direct_path(ctx, n):
    m = rand_struct(AFF, n, n + 2)
    assert ctx.reduce(AFF3, ctx.vector(m)).tobytes() == oracle.skel_reduce(AFF3, m).tobytes()


def test_reduce_closed_form_matrix_power(ctx):
    n = 1_000_003
    m = np.zeros(n, M2)
    m["a"], m["b"], m["d"] = 1, 1, 1
    r = ctx.reduce(MAT_U, ctx.vector(m))
    assert (int(r["a"]), int(r["b"]), int(r["c"]), int(r["d"])) == (1, n, 0, 1)


def test_listing1_dot_product(ctx):
    n = 1 << 20
    a, b = si.uniform_f32(n, 1), si.uniform_f32(n, 2)
    A, B = ctx.vector(a), ctx.vector(b)
    prod = ctx.vector(n=n, dtype=np.float32)
    ctx.zip(MULT_F32, A, B, prod)
    got = float(ctx.reduce(SUM_F32, prod))
    p = oracle.skel_zip(MULT_F32, a, b, np.float32)
    assert_sum_close(got, p)


def test_reduce_to_vector(ctx):
    x = si.uniform_int01(100_000, 1)
    r = ctx.vector(n=1, dtype=np.int32)
    ctx.reduce_to(SUM_I32, ctx.vector(x), r)
    assert int(r.download()[0]) == int(x.sum())


# ---- Scan -----------------------------------------------------------------------
def assert_scan_close(got, x):
    want, ab = oracle.exscan_f32_exact(x)
    err = np.abs(got.astype(np.float64) - want.astype(np.float64))
    tol = 1e-5 * ab + 1e-30
    bad = np.nonzero(err > tol)[0]
    assert bad.size == 0, (bad[:5], got[bad[:5]], want[bad[:5]])


@pytest.mark.parametrize("n", SIZES)
def test_scan_sum_f32(ctx, n):
    x = si.uniform_f32(n, 31 + n % 7)
    out = ctx.vector(n=n, dtype=np.float32)
    ctx.scan(SUM_F32, ctx.vector(x), out, np.float32(0))
    got = out.download()
    assert got[0] == 0.0
    assert_scan_close(got, x)


@pytest.mark.parametrize("n", SIGNED_SIZES)
@pytest.mark.parametrize("gen", ["signed", "cancel"])
def test_scan_sum_f32_signed(ctx, n, gen):
    x = (si.uniform_signed_f32 if gen == "signed" else si.cancellation_f32)(n, 50 + n % 7)
    out = ctx.vector(n=n, dtype=np.float32)
    ctx.scan(SUM_F32, ctx.vector(x), out, np.float32(0))
    got = out.download()
    assert got[0] == 0.0
    assert_scan_close(got, x)


@pytest.mark.parametrize("n", SIZES)
def test_scan_sum_i32_exact(ctx, n):
    x = si.uniform_int01(n, 8)
    out = ctx.vector(n=n, dtype=np.int32)
    ctx.scan(SUM_I32, ctx.vector(x), out, np.int32(0))
    assert np.array_equal(out.download(), oracle.skel_scan(SUM_I32, x, 0))


def test_scan_identity_is_the_given_one(ctx):
    out = ctx.vector(n=5, dtype=np.int32)
    ctx.scan(SUM_I32, ctx.vector(np.arange(5, dtype=np.int32)), out, np.int32(7))
    assert out.download().tolist() == [7, 7, 8, 10, 13]


@pytest.mark.parametrize("n", [1, 2, 33, 8192, 8193, 3 * 8192 + 5, 300_001])
def test_scan_noncommutative_16B(ctx, n):
    m = rand_struct(M2, n, 100 + n)
    ident = np.zeros(1, M2)
    ident["a"], ident["d"] = 1, 1
    out = ctx.vector(n=n, dtype=M2)
    ctx.scan(MAT_U, ctx.vector(m), out, ident[0])
    assert out.download().tobytes() == oracle.skel_scan(MAT_U, m, ident[0]).tobytes()


@pytest.mark.parametrize("n", [3, 16384, 16385, 100_003])
def test_scan_noncommutative_8B(ctx, n):
    m = rand_struct(A2, n, 200 + n)
    ident = np.zeros(1, A2)
    ident["a"] = 1
    out = ctx.vector(n=n, dtype=A2)
    ctx.scan(AFF2, ctx.vector(m), out, ident[0])
    assert out.download().tobytes() == oracle.skel_scan(AFF2, m, ident[0]).tobytes()


@pytest.mark.parametrize("n", [3, 5461, 5462, 60_001])
def test_scan_noncommutative_12B_direct_path(ctx, n):
    m = rand_struct(AFF, n, 300 + n)
    ident = np.zeros(1, AFF)
    ident["a"] = 1
    out = ctx.vector(n=n, dtype=AFF)
    ctx.scan(AFF3, ctx.vector(m), out, ident[0])
    assert out.download().tobytes() == oracle.skel_scan(AFF3, m, ident[0]).tobytes()


def test_scan_inplace_and_repeated_launches(ctx):
    x = si.uniform_int01(500_001, 4)
    v = ctx.vector(x)
    ctx.scan(SUM_I32, v, v, np.int32(0))  # in place
    assert np.array_equal(v.download(), oracle.skel_scan(SUM_I32, x, 0))
    # many launches back to back: epochs and tickets must reset correctly
    out = ctx.vector(n=x.size, dtype=np.int32)
    vx = ctx.vector(x)
    for _ in range(20):
        ctx.scan(SUM_I32, vx, out, np.int32(0))
    assert np.array_equal(out.download(), oracle.skel_scan(SUM_I32, x, 0))


def test_scan_last_plus_x_equals_reduce(ctx):
    x = si.uniform_u32(1_000_001, 6)
    src = "unsigned add(unsigned a, unsigned b){ return a + b; }"
    out = ctx.vector(n=x.size, dtype=np.uint32)
    vx = ctx.vector(x)
    ctx.scan(src, vx, out, np.uint32(0))
    assert np.uint32(out.download()[-1] + x[-1]) == ctx.reduce(src, vx)


BIG = """
struct Big { double a[3]; unsigned n; unsigned p; };   /* 32-byte element, direct path */
/* .a: exact float64 sums; (.n, .p): base-3 Horner digits mod 2^32 -- associative, not commutative */
Big bsum(Big x, Big y) { Big r; for (int i = 0; i < 3; ++i) r.a[i] = x.a[i] + y.a[i]; r.n = x.n * y.p + y.n; r.p = x.p * y.p; return r; }
"""
BIG_DT = np.dtype([("a", np.float64, (3,)), ("n", np.uint32), ("p", np.uint32)])


@pytest.mark.parametrize("n", [1, 100, 5000, 200_003])
def test_32byte_elements_reduce_scan(ctx, n):
    g = np.random.default_rng(n)
    x = np.zeros(n, BIG_DT)
    x["a"] = g.integers(0, 1000, (n, 3)).astype(np.float64)  # exact in float64: any order
    x["n"] = g.integers(0, 3, n).astype(np.uint32)
    x["p"] = 3
    r = ctx.reduce(BIG, ctx.vector(x))
    want = oracle.skel_reduce(BIG, x)
    assert r.tobytes() == want.tobytes()  # .n is order-sensitive, .a exact
    ident = np.zeros(1, BIG_DT)
    ident["p"] = 1
    out = ctx.vector(n=n, dtype=BIG_DT)
    ctx.scan(BIG, ctx.vector(x), out, ident[0])
    assert out.download().tobytes() == oracle.skel_scan(BIG, x, ident[0]).tobytes()


@pytest.mark.parametrize("n", [3, 16385, 1_000_001])
def test_double_reduce_scan(ctx, n):
    src = "double add(double a, double b){ return a + b; }"
    x = si.uniform_f32(n, 4).astype(np.float64)
    r = float(ctx.reduce(src, ctx.vector(x)))
    assert abs(r - float(np.sum(x))) <= 1e-12 * float(np.sum(np.abs(x)))
    out = ctx.vector(n=n, dtype=np.float64)
    ctx.scan(src, ctx.vector(x), out, np.float64(0))
    want = oracle.skel_scan(src, x, 0.0)  # left-to-right float64 prefix
    got = out.download()
    assert np.all(np.abs(got - want) <= 1e-12 * np.concatenate([[0], np.cumsum(np.abs(x))[:-1]]) + 1e-300)


@pytest.mark.parametrize("n", [(1 << 22) + 5, 1 << 24])
def test_map_zip_grid_policy_trials_bit_identical(n, tmp_path):
    """The element-wise grid policy is chosen per module and size class by timing
    the three candidates on the first launches (K1/K2): every
    launch -- trials of each policy (incl. the scalar one-element-per-thread
    path) and the decided one -- must give the same bits."""
    with skel.Context(1) as c:
        c.set_cache_dir(str(tmp_path))  # no decisions persisted by earlier processes: trials run
        x, y = si.uniform_f32(n, 11), si.uniform_f32(n, 12)
        vx, vy = c.vector(x), c.vector(y)
        want_m = oracle.skel_map(MAP_F32, x, np.float32)
        want_z = oracle.skel_zip(SAXPY_F32, x, y, np.float32, args=[np.float32(2.5)])
        for _ in range(7):
            vm = c.vector(n=n, dtype=np.float32)
            vz = c.vector(n=n, dtype=np.float32)
            c.map(MAP_F32, vx, vm)
            c.zip(SAXPY_F32, vx, vy, vz, args=[np.float32(2.5)])
            assert np.array_equal(vm.download(), want_m)
            assert np.array_equal(vz.download(), want_z)
            vm.destroy()
            vz.destroy()


_POLICY_CHILD = r"""
import sys, numpy as np
sys.path.insert(0, {root!r})
import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import MAP_F32
with skel.Context(1) as c:
    c.set_cache_dir({cache!r})
    x = si.uniform_f32(1 << 22, 3)
    vx, vm = c.vector(x), c.vector(n=x.size, dtype=np.float32)
    c.map(MAP_F32, vx, vm)
    c.sync()
    print("LAUNCHES", c.stats()["kernel_launches"])
"""


def test_grid_policy_decisions_persist_across_processes(tmp_path):
    """A decided grid policy is written next to the cached cubin (<key>.policy)
    and a later process takes it without trials (one launch instead of the
    trial launches); SKEL_POLICY_CACHE=0 turns the file off."""
    import os, re, subprocess, sys
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    code = _POLICY_CHILD.format(root=root, cache=str(tmp_path))

    def run(env_extra):
        env = dict(os.environ, SKEL_LOG="1", **env_extra)
        r = subprocess.run([sys.executable, "-c", code], capture_output=True, text=True, env=env, timeout=300)
        assert r.returncode == 0, r.stderr
        return int(re.search(r"LAUNCHES (\d+)", r.stdout).group(1)), r.stderr.count("grid policy")

    n1, t1 = run({})
    assert t1 == 1 and n1 > 1  # trials, then the launch
    files = [f for f in os.listdir(tmp_path) if f.endswith(".policy")]
    assert len(files) == 1
    tag, cls, _h, pol = open(tmp_path / files[0]).read().split()
    assert tag.startswith("cc") and int(pol) in range(5) and int(cls) >= 18
    n2, t2 = run({})
    assert (n2, t2) == (1, 0)  # decision from the file, no trials
    n3, t3 = run({"SKEL_POLICY_CACHE": "0"})
    assert t3 == 1 and n3 > 1


IDX_I64 = "long long poly(long long i, long long k){ return i * i - k * i + 7; }"


@pytest.mark.parametrize("D,dist", [(1, None), (2, skel.BLOCK), (3, skel.BLOCK), (3, skel.COPY), (2, skel.SINGLE)])
@pytest.mark.parametrize("n", [1, 5, 4097, (1 << 20) + 3])
def test_index_map_is_map_over_the_index_vector(D, dist, n):
    """NEXT-4: map_index(f, n) equals Map(f) over [0, 1, ..., n-1] (eq. (1)), with
    global indices under a block distribution of the output."""
    want = oracle.skel_map(IDX_I64, np.arange(n, dtype=np.int64), np.int64, args=[np.int64(5)])
    with skel.Context(D) as c:
        out = c.vector(n=n, dtype=np.int64)
        if dist is not None:
            out.set_distribution(dist)
        c.map_index(IDX_I64, n, out, args=[np.int64(5)])
        assert np.array_equal(out.download(), want)


def test_void_index_map_side_effects():
    n = 10_007
    with skel.Context(2) as c:
        acc = c.vector(np.zeros(n, np.int32))
        acc.set_distribution(skel.COPY)
        c.map_index("void touch(int i, int* a){ a[i] += i % 5 + 1; }", n, None, args=[acc])
        acc.mark_device_modified()
        acc.set_distribution(skel.BLOCK, skel.COMBINE_ADD)
        assert np.array_equal(acc.download(), (np.arange(n) % 5 + 1).astype(np.int32))


@pytest.mark.parametrize("n", [(1 << 21) + 5, 3_000_017])
def test_small_paths_with_double_tiles_i32(ctx, n):
    """Between 8 and 16 MiB the Reduce takes its small-vector path with
    double-size tiles and the Scan (above its 8 MiB switch point) the
    persistent path: integer results bit-exact."""
    x = si.uniform_int01(n, 21)
    vx = ctx.vector(x)
    assert int(ctx.reduce(SUM_I32, vx)) == int(x.astype(np.int64).sum())
    out = ctx.vector(n=n, dtype=np.int32)
    ctx.scan(SUM_I32, vx, out, np.int32(0))
    assert np.array_equal(out.download(), oracle.skel_scan(SUM_I32, x, 0))


def test_small_paths_with_double_tiles_noncommutative_16B(ctx):
    n = 700_001  # 11.2 MB of 16-byte elements
    m = rand_struct(M2, n, 77)
    assert ctx.reduce(MAT_U, ctx.vector(m)).tobytes() == oracle.skel_reduce(MAT_U, m).tobytes()
    ident = np.zeros(1, M2)
    ident["a"], ident["d"] = 1, 1
    out = ctx.vector(n=n, dtype=M2)
    ctx.scan(MAT_U, ctx.vector(m), out, ident[0])
    assert out.download().tobytes() == oracle.skel_scan(MAT_U, m, ident[0]).tobytes()
