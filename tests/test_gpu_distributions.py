"""Distributions and multi-device skeletons (§III-D, Listing 4) on D
logical devices.  With one physical GPU the logical devices are "virtual"
(skel_init(D) maps them all onto GPU 0; exchanges use the library's own
copy/combine kernels).  Every result is checked against the oracle's pure
distribution model and skeleton definitions; integer results must be
bit-identical to D = 1."""
import itertools

import numpy as np
import pytest

import oracle
import skel_inputs as si
from oracle import distribution as odist
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import MAP_I32, SAXPY_F32, SUM_F32, SUM_I32

pytestmark = pytest.mark.gpu

DISTS = [skel.SINGLE, skel.BLOCK, skel.COPY]
NAMES = {skel.SINGLE: odist.SINGLE, skel.BLOCK: odist.BLOCK, skel.COPY: odist.COPY}
IDENT_I32 = "int ident(int x){ return x; }"


def on_devices(ctx, x, dist):
    """A vector whose data live on the devices under `dist` (not just the host)."""
    v = ctx.vector(x)
    v.set_distribution(dist)  # lazy: host-only data
    w = ctx.vector(n=x.size, dtype=x.dtype)
    ctx.map(IDENT_I32, v, w)  # w: device-valid, distributed like v
    assert w.distribution == dist
    return w


@pytest.mark.parametrize("D", [2, 3, 4, 8])
@pytest.mark.parametrize("n", [1, 5, 37, 4099, 100_003])
def test_every_transition_preserves_the_vector(D, n):
    x = si.uniform_i32(n, n)
    with skel.Context(D) as ctx:
        for a, b in itertools.product(DISTS, DISTS):
            w = on_devices(ctx, x, a)
            w.set_distribution(b)
            assert w.distribution == b
            assert np.array_equal(w.download(), x), (a, b)
            # parts follow the planner
            for d in range(D):
                lo, hi = w.part(d)
                if b == skel.BLOCK:
                    assert (lo, hi) == odist.part_range(n, D, d)


@pytest.mark.parametrize("D", [2, 4, 8])
def test_copy_to_block_add_of_equal_copies(D):
    x = np.arange(10_001, dtype=np.float32)
    with skel.Context(D) as ctx:
        v = ctx.vector(x)
        v.set_distribution(skel.COPY)
        w = ctx.vector(n=x.size, dtype=np.float32)
        ctx.map("float id(float x){ return x; }", v, w)
        w.set_distribution(skel.BLOCK, skel.COMBINE_ADD)
        model = odist.redistribute(odist.distribute(x, odist.COPY, D), odist.COPY, odist.BLOCK, "add")
        assert np.array_equal(w.download(), np.concatenate(model))


@pytest.mark.parametrize("D", [2, 3, 4, 8])
@pytest.mark.parametrize("dst", [skel.BLOCK, skel.SINGLE, skel.COPY])
def test_combine_of_diverged_copies(D, dst):
    """Each device writes its own block's indices into its own copy (side-effect
    Map); the combine then merges the D different copies."""
    n = 50_001
    base = np.arange(n, dtype=np.int32) % 1000
    mark = "void mark(int i, int* c){ c[i] += 1 + i % 7; }"
    with skel.Context(D) as ctx:
        c = ctx.vector(base)
        c.set_distribution(skel.COPY)
        idx = ctx.vector(np.arange(n, dtype=np.int32))
        idx.set_distribution(skel.BLOCK)
        ctx.map(mark, idx, None, args=[c])
        c.mark_device_modified()
        c.set_distribution(dst, skel.COMBINE_ADD)
        copies = []
        for d in range(D):
            cd = base.copy()
            lo, hi = odist.part_range(n, D, d)
            cd[lo:hi] += 1 + np.arange(lo, hi) % 7
            copies.append(cd)
        model = odist.redistribute(copies, odist.COPY, NAMES[dst], "add")
        assert np.array_equal(c.download(), odist.gather(model, NAMES[dst]))


@pytest.mark.parametrize("D", [2, 3, 4, 8])
def test_copy_to_block_without_combine_keeps_local_slices(D):
    n = 999
    mark = "void mark(int i, int* c){ c[i] = 5; }"
    with skel.Context(D) as ctx:
        c = ctx.vector(np.zeros(n, np.int32))
        c.set_distribution(skel.COPY)
        idx = ctx.vector(np.arange(n, dtype=np.int32))
        idx.set_distribution(skel.BLOCK)
        ctx.map(mark, idx, None, args=[c])
        c.mark_device_modified()
        c.set_distribution(skel.BLOCK)
        # each device wrote exactly its own slice, so the local slices are all 5
        assert (c.download() == 5).all()


@pytest.mark.parametrize("D", [2, 3, 4, 8])
@pytest.mark.parametrize("n", [1, 3, 16385, 1_000_003])
def test_cross_device_reduce_and_scan_int_bit_identical(D, n):
    x = si.uniform_int01(n, n + D)
    want_r = int(oracle.skel_reduce(SUM_I32, x))
    want_s = oracle.skel_scan(SUM_I32, x, 0)
    with skel.Context(D) as ctx:
        v = ctx.vector(x)
        v.set_distribution(skel.BLOCK)
        assert int(ctx.reduce(SUM_I32, v)) == want_r
        out = ctx.vector(n=n, dtype=np.int32)
        ctx.scan(SUM_I32, v, out, np.int32(0))
        assert out.distribution == skel.BLOCK
        assert np.array_equal(out.download(), want_s)


@pytest.mark.parametrize("D", [2, 4, 8])
def test_cross_device_noncommutative_order(D):
    src = """
    struct M2 { unsigned a, b, c, d; };
    M2 matmul(M2 x, M2 y) {
      M2 r;
      r.a = x.a*y.a + x.b*y.c;  r.b = x.a*y.b + x.b*y.d;
      r.c = x.c*y.a + x.d*y.c;  r.d = x.c*y.b + x.d*y.d;
      return r;
    }"""
    M2 = np.dtype([("a", np.uint32), ("b", np.uint32), ("c", np.uint32), ("d", np.uint32)])
    n = 123_457
    g = np.random.default_rng(D)
    m = np.zeros(n, M2)
    for k in "abcd":
        m[k] = g.integers(0, 1 << 32, n, dtype=np.uint64).astype(np.uint32)
    ident = np.zeros(1, M2)
    ident["a"], ident["d"] = 1, 1
    with skel.Context(D) as ctx:
        v = ctx.vector(m)
        v.set_distribution(skel.BLOCK)
        assert ctx.reduce(src, v).tobytes() == oracle.skel_reduce(src, m).tobytes()
        out = ctx.vector(n=n, dtype=M2)
        ctx.scan(src, v, out, ident[0])
        assert out.download().tobytes() == oracle.skel_scan(src, m, ident[0]).tobytes()


@pytest.mark.parametrize("D", [2, 4])
@pytest.mark.parametrize("gen", ["uniform", "signed", "cancel"])
@pytest.mark.parametrize("n", [(1 << 20) + 77, (1 << 26) + 3])
def test_cross_device_float_reduce_scan_within_tolerance(D, gen, n):
    x = {"uniform": si.uniform_f32, "signed": si.uniform_signed_f32, "cancel": si.cancellation_f32}[gen](n, 9)
    with skel.Context(D) as ctx:
        v = ctx.vector(x)
        v.set_distribution(skel.BLOCK)
        r = float(ctx.reduce(SUM_F32, v))
        assert abs(r - oracle.sum_f32_exact(x)) <= 1e-5 * oracle.abssum_f32(x)
        out = ctx.vector(n=n, dtype=np.float32)
        ctx.scan(SUM_F32, v, out, np.float32(0))
        want, ab = oracle.exscan_f32_exact(x)
        assert np.all(np.abs(out.download().astype(np.float64) - want) <= 1e-5 * ab)


@pytest.mark.parametrize("D", [2, 3, 8])
def test_zip_brings_b_to_a_distribution(D):
    n = 77_777
    x, y = si.uniform_f32(n, 1), si.uniform_f32(n, 2)
    with skel.Context(D) as ctx:
        a = ctx.vector(x)
        a.set_distribution(skel.BLOCK)
        b = ctx.vector(y)
        b.set_distribution(skel.COPY)
        out = ctx.vector(n=n, dtype=np.float32)
        ctx.zip(SAXPY_F32, a, b, out, args=[np.float32(2.5)])
        assert b.distribution == skel.BLOCK and out.distribution == skel.BLOCK
        assert np.array_equal(out.download(), oracle.skel_zip(SAXPY_F32, x, y, np.float32,
                                                              args=[np.float32(2.5)]))


@pytest.mark.parametrize("dist", DISTS)
def test_map_under_each_distribution(dist):
    x = si.uniform_i32(30_001, 5)
    with skel.Context(4) as ctx:
        v = ctx.vector(x)
        v.set_distribution(dist)
        out = ctx.vector(n=x.size, dtype=np.int32)
        ctx.map(MAP_I32, v, out)
        assert out.distribution == dist
        assert np.array_equal(out.download(), oracle.skel_map(MAP_I32, x, np.int32))
        # copies are computed redundantly: every device holds the full result
        if dist == skel.COPY:
            for li in range(4):
                assert out.device_ptr(li)[1] == x.size


@pytest.mark.parametrize("D", [3, 5, 7])
@pytest.mark.parametrize("n", [1001, 70_003])
def test_skeletons_on_unaligned_block_views(D, n):
    """copy -> block keeps each device's part inside its full buffer at offset
    k*ceil(n/D) (no data movement); for these (n, D) the parts start at
    addresses that are not 16-byte aligned, which must route every skeleton to
    its unaligned path."""
    xi = si.uniform_int01(n, 1)
    xf = si.uniform_f32(n, 2)
    with skel.Context(D) as ctx:
        vi = ctx.vector(xi)
        vi.set_distribution(skel.COPY)
        wi = ctx.vector(n=n, dtype=np.int32)
        ctx.map(IDENT_I32, vi, wi)  # device-valid copies
        wi.set_distribution(skel.BLOCK)  # local slices, aliased
        assert int(ctx.reduce(SUM_I32, wi)) == int(xi.sum())
        out = ctx.vector(n=n, dtype=np.int32)
        ctx.scan(SUM_I32, wi, out, np.int32(0))
        assert np.array_equal(out.download(), oracle.skel_scan(SUM_I32, xi, 0))
        m = ctx.vector(n=n, dtype=np.int32)
        ctx.map(MAP_I32, wi, m)
        assert np.array_equal(m.download(), oracle.skel_map(MAP_I32, xi, np.int32))
        vf = ctx.vector(xf)
        vf.set_distribution(skel.COPY)
        wf = ctx.vector(n=n, dtype=np.float32)
        ctx.map("float id(float x){ return x; }", vf, wf)
        wf.set_distribution(skel.BLOCK)
        z = ctx.vector(n=n, dtype=np.float32)
        ctx.zip(SAXPY_F32, wf, wf, z, args=[np.float32(2.5)])
        assert np.array_equal(z.download(), oracle.skel_zip(SAXPY_F32, xf, xf, np.float32, args=[np.float32(2.5)]))


def test_more_devices_than_elements():
    x = np.arange(3, dtype=np.int32)
    with skel.Context(8) as ctx:
        v = ctx.vector(x)
        v.set_distribution(skel.BLOCK)
        assert int(ctx.reduce(SUM_I32, v)) == 3
        out = ctx.vector(n=3, dtype=np.int32)
        ctx.scan(SUM_I32, v, out, np.int32(0))
        assert out.download().tolist() == [0, 0, 1]
        v.set_distribution(skel.COPY)
        v.set_distribution(skel.SINGLE)
        assert v.download().tolist() == [0, 1, 2]


# NEXT-2: user-defined combine functions (skel_vector_set_distribution_fn)
MAX_I32 = "int mx(int a, int b){ return a > b ? a : b; }"
AFF2_SRC = """
struct A2 { unsigned a, b; };
A2 comp2(A2 f, A2 g) { A2 r; r.a = f.a * g.a; r.b = f.b * g.a + g.b; return r; }
"""
A2 = np.dtype([("a", np.uint32), ("b", np.uint32)])


def diverged_copies_i32(ctx, base, D):
    """copy d = base with part d overwritten by a side-effect Map (device d's events)"""
    n = base.size
    c = ctx.vector(base)
    c.set_distribution(skel.COPY)
    idx = ctx.vector(np.arange(n, dtype=np.int32))
    idx.set_distribution(skel.BLOCK)
    ctx.map("void mark(int i, int* c){ c[i] = (i * 7919) % 1000 - 500; }", idx, None, args=[c])
    c.mark_device_modified()
    copies = []
    for d in range(D):
        cd = base.copy()
        lo, hi = odist.part_range(n, D, d)
        cd[lo:hi] = (np.arange(lo, hi) * 7919) % 1000 - 500
        copies.append(cd)
    return c, copies


@pytest.mark.parametrize("D", [2, 3, 4])
@pytest.mark.parametrize("dst", [skel.BLOCK, skel.SINGLE, skel.COPY])
def test_user_combine_max_of_diverged_copies(D, dst):
    n = 30_011
    base = (np.arange(n, dtype=np.int32) % 613) - 300
    with skel.Context(D) as ctx:
        c, copies = diverged_copies_i32(ctx, base, D)
        c.set_distribution(dst, MAX_I32)
        assert c.distribution == dst
        f = lambda a, b: oracle.skel_zip(MAX_I32, a, b, np.int32)
        model = odist.redistribute(copies, odist.COPY, NAMES[dst], f)
        assert np.array_equal(c.download(), odist.gather(model, NAMES[dst]))


@pytest.mark.parametrize("D", [2, 3, 4])
@pytest.mark.parametrize("dst", [skel.BLOCK, skel.SINGLE])
def test_user_combine_noncommutative_struct_in_device_order(D, dst):
    """8-byte affine maps composed across the copies: only the device order
    0..D-1 gives the oracle's result (the function is not commutative)."""
    n = 4099
    g = np.random.default_rng(7)
    base = np.zeros(n, A2)
    base["a"] = g.integers(1, 1 << 16, n)
    base["b"] = g.integers(0, 1 << 16, n)
    mk = """
struct A2 { unsigned a, b; };
void mk(int i, A2* c){ c[i].a = 2u * (unsigned)i + 3u; c[i].b = (unsigned)i * 40503u; }
"""
    with skel.Context(D) as ctx:
        c = ctx.vector(base)
        c.set_distribution(skel.COPY)
        idx = ctx.vector(np.arange(n, dtype=np.int32))
        idx.set_distribution(skel.BLOCK)
        ctx.map(mk, idx, None, args=[c])
        c.mark_device_modified()
        copies = []
        for d in range(D):
            cd = base.copy()
            lo, hi = odist.part_range(n, D, d)
            i = np.arange(lo, hi, dtype=np.uint64)
            cd["a"][lo:hi] = (2 * i + 3).astype(np.uint32)
            cd["b"][lo:hi] = ((i * 40503) % (1 << 32)).astype(np.uint32)
            copies.append(cd)
        c.set_distribution(dst, AFF2_SRC)
        f = lambda a, b: oracle.skel_zip(AFF2_SRC, a, b, A2)
        want = odist.gather(odist.redistribute(copies, odist.COPY, NAMES[dst], f), NAMES[dst])
        assert c.download().tobytes() == want.tobytes()
        rev = odist.gather(odist.redistribute(copies[::-1], odist.COPY, NAMES[dst], f), NAMES[dst])
        assert want.tobytes() != rev.tobytes()  # the order matters for this data


def test_user_combine_errors():
    with skel.Context(2) as ctx:
        v = ctx.vector(np.arange(10, dtype=np.int32))
        v.set_distribution(skel.BLOCK)
        with pytest.raises(skel.SkelError) as e:
            v.set_distribution(skel.BLOCK, MAX_I32)  # not copy-distributed
        assert e.value.status == 8  # SKEL_ERR_STATE
        v.set_distribution(skel.COPY)
        with pytest.raises(skel.SkelError) as e:
            v.set_distribution(skel.BLOCK, "double f(double a, double b){ return a + b; }")
        assert e.value.status == 3  # SKEL_ERR_TYPE
        with pytest.raises(skel.SkelError) as e:
            v.set_distribution(skel.BLOCK, "int f(int a, int b, int k){ return a + b + k; }")
        assert e.value.status == 3  # SKEL_ERR_TYPE


@pytest.mark.parametrize("D", [2, 3, 8])
def test_cross_device_reduce_single_pass(D):
    """A block-distributed Reduce over in-process devices folds the device
    results inside the Reduce kernels (the last device to finish folds them
    in device order): counted by xdev_reduces, exact for a
    non-commutative operator, its arrival counter reset for the next Reduce
    (40 in a row, sizes on both the small and the TMA path) and across CUDA
    graph replays of a reduce_to."""
    src = """
    struct A { unsigned m, c; };
    A affine(A x, A y) { A r; r.m = x.m * y.m; r.c = x.c * y.m + y.c; return r; }"""
    AF = np.dtype([("m", np.uint32), ("c", np.uint32)])
    g = np.random.default_rng(D)
    with skel.Context(D) as ctx:
        x0 = ctx.stats()["xdev_reduces"]
        for i in range(40):
            n = [7, 1000, 300_007, 5_000_011][i % 4]
            a = np.zeros(n, AF)
            a["m"] = g.integers(0, 1 << 32, n, dtype=np.uint64).astype(np.uint32)
            a["c"] = g.integers(0, 1 << 32, n, dtype=np.uint64).astype(np.uint32)
            v = ctx.vector(a)
            v.set_distribution(skel.BLOCK)
            assert ctx.reduce(src, v).tobytes() == oracle.skel_reduce(src, a).tobytes(), (i, n)
            v.destroy()
        assert ctx.stats()["xdev_reduces"] - x0 == 40
        x = si.uniform_int01(2_000_003, 77)
        v = ctx.vector(x)
        v.set_distribution(skel.BLOCK)
        r = ctx.vector(n=1, dtype=np.int32)
        ctx.reduce_to(SUM_I32, v, r)  # eager first: workspaces are sized outside the capture
        ctx.sync()
        gr = ctx.capture(lambda: ctx.reduce_to(SUM_I32, v, r))
        for _ in range(20):
            gr.launch()
            ctx.sync()
            r.mark_device_modified()
            assert int(r.download()[0]) == int(x.sum())
        gr.destroy()


def test_cross_device_reduce_single_pass_matches_the_two_step_exchange():
    """SKEL_XDEV_REDUCE=0 (gather of the device results + fold launches) and
    the single pass give bit-identical integer and ordered results."""
    import subprocess
    import sys
    from pathlib import Path
    code = r'''
import sys; sys.path.insert(0, ".")
import numpy as np, skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import SUM_I32
x = si.uniform_int01(1_000_003, 5)
with skel.Context(4) as ctx:
    v = ctx.vector(x); v.set_distribution(skel.BLOCK)
    o = ctx.vector(n=x.size, dtype=np.int32)
    ctx.scan(SUM_I32, v, o, np.int32(0))
    print(int(ctx.reduce(SUM_I32, v)), int(o.download()[-1]), ctx.stats()["xdev_reduces"])
'''
    root = Path(__file__).resolve().parents[1]
    outs = {}
    for flag in ("0", "1"):
        env = dict(__import__("os").environ, SKEL_XDEV_REDUCE=flag)
        r = subprocess.run([sys.executable, "-c", code], capture_output=True, text=True, cwd=str(root), env=env,
                           timeout=300)
        assert r.returncode == 0, r.stderr[-2000:]
        outs[flag] = r.stdout.split()
    assert outs["0"][:2] == outs["1"][:2]
    assert outs["0"][2] == "0" and int(outs["1"][2]) >= 2  # the Scan's device results come through it too
