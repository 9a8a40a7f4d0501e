"""Parity at BASELINE.json's full sweep size (configs[1]: 2^30 float32 and
int32 elements) in the launch configuration bench.py times (one B200, single
distribution, the same skeleton functions).  Outputs are checked on samples
the oracle computes one by one (sequential float64 prefix sums evaluated at
the sampled positions), plus whole-vector properties."""
import numpy as np
import pytest

import oracle
import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import MAP_F32, SAXPY_F32, SUM_F32, SUM_I32

pytestmark = pytest.mark.gpu

N = 1 << 30


@pytest.fixture(scope="module")
def ctx():
    c = skel.Context(1)
    yield c
    c.close()


@pytest.fixture(scope="module")
def data():
    return si.uniform_f32(N, 20110516), si.uniform_f32(N, 20110517)


def sample_idx(n, k=200_000, seed=0):
    g = np.random.default_rng(seed)
    idx = np.unique(np.concatenate([g.integers(0, n, k), np.arange(8), n - 1 - np.arange(8),
                                    np.arange(0, n, 16384 * 148)]))
    return idx[idx < n]


def test_full_size_float_step(ctx, data):
    x, y = data
    X, Y = ctx.vector(x), ctx.vector(y)
    m = ctx.vector(n=N, dtype=np.float32)
    z = ctx.vector(n=N, dtype=np.float32)
    s = ctx.vector(n=N, dtype=np.float32)
    ctx.map(MAP_F32, X, m)
    ctx.zip(SAXPY_F32, X, Y, z, args=[np.float32(2.5)])
    r = float(ctx.reduce(SUM_F32, X))
    ctx.scan(SUM_F32, X, s, np.float32(0))
    idx = sample_idx(N)
    # Map / Zip: bit-exact on the samples
    mg = m.download()
    assert np.array_equal(mg[idx], oracle.skel_map(MAP_F32, x[idx], np.float32))
    del mg
    zg = z.download()
    assert np.array_equal(zg[idx], oracle.skel_zip(SAXPY_F32, x[idx], y[idx], np.float32,
                                                   args=[np.float32(2.5)]))
    del zg
    # Reduce: normwise 1e-5 against the exact sum
    assert abs(r - oracle.sum_f32_exact(x)) <= 1e-5 * oracle.abssum_f32(x)
    # Scan: per element |y_i - exact_i| <= 1e-5 * sum_{j<i} |x_j|
    sg = s.download()
    sidx, pre, ab = oracle.exscan_f32_sampled(x, idx)
    err = np.abs(sg[sidx].astype(np.float64) - pre)
    assert np.all(err <= 1e-5 * ab), float(np.max(err / np.maximum(ab, 1e-30)))
    # the relative error actually reached (reported by the assertion message above)
    assert float(np.max(err[1:] / ab[1:])) < 1e-5


def test_full_size_int_scan_and_reduce(ctx):
    x = si.uniform_int01(N, 7)
    X = ctx.vector(x)
    out = ctx.vector(n=N, dtype=np.int32)
    ctx.scan(SUM_I32, X, out, np.int32(0))
    total = int(ctx.reduce(SUM_I32, X))
    assert total == int(x.sum(dtype=np.int64))
    g = out.download()
    assert np.array_equal(g, oracle.skel_scan(SUM_I32, x, 0))  # whole vector, bit-exact
    assert int(g[-1]) + int(x[-1]) == total


@pytest.mark.parametrize("gen", ["signed", "cancel"])
def test_full_size_signed_reduce_scan(ctx, gen):
    """Signed data (U[-1,1)) and catastrophic cancellation ([+-2^24, u, -+2^24, u'])
    at 2^30 through the persistent Scan and the TMA Reduce."""
    x = (si.uniform_signed_f32 if gen == "signed" else si.cancellation_f32)(N, 20110600)
    X = ctx.vector(x)
    s = ctx.vector(n=N, dtype=np.float32)
    r = float(ctx.reduce(SUM_F32, X))
    assert abs(r - oracle.sum_f32_exact(x)) <= 1e-5 * oracle.abssum_f32(x)
    ctx.scan(SUM_F32, X, s, np.float32(0))
    sg = s.download()
    idx = sample_idx(N, seed=3)
    sidx, pre, ab = oracle.exscan_f32_sampled(x, idx)
    err = np.abs(sg[sidx].astype(np.float64) - pre)
    assert np.all(err <= 1e-5 * ab), float(np.max(err[1:] / ab[1:]))
