"""Forward progress of the persistent Scan.

The persistent Scan's window for CTA c waits on aggregates published by
higher-index CTAs of the previous slice, so its whole grid must be resident at
once (eq. (4), computed by a single-pass grid).  The library
launches it cooperatively (co-residency guaranteed or the launch refused ->
two short launches) and chains the persistent Scans of logical devices that
share one GPU.  These tests force the persistent path (SKEL_SCAN_SMALL_MAX=0)
into the configurations that could interleave two grids or starve one:

* 8 virtual devices on one GPU, copy distribution: 8 full-vector Scans at once;
* a second context keeping every SM busy with a long-running Map while the
  Scan is launched on another stream.

Each runs in a subprocess under a timeout, so a hang fails the test instead of
hanging the suite; results are compared with the oracle (int32 bit-exact)."""
import os
import subprocess
import sys
import textwrap

import pytest

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))

PRELUDE = textwrap.dedent("""
    import sys
    sys.path.insert(0, %r)
    import numpy as np
    import oracle
    import skel_inputs as si
    from paper_conf_ipps_steuwerkg11_b200 import skel
    from paper_conf_ipps_steuwerkg11_b200.workloads import SUM_I32
""" % ROOT)


def run(body: str, timeout: int = 240):
    env = dict(os.environ, SKEL_SCAN_SMALL_MAX="0")
    r = subprocess.run([sys.executable, "-c", PRELUDE + textwrap.dedent(body)], env=env, cwd=ROOT,
                       capture_output=True, text=True, timeout=timeout)
    assert r.returncode == 0, r.stdout[-2000:] + r.stderr[-3000:]
    return r.stdout


def test_eight_virtual_devices_concurrent_persistent_scans():
    out = run("""
        n = (1 << 22) + 5
        x = si.uniform_int01(n, 77)
        want = oracle.skel_scan(SUM_I32, x, 0)
        with skel.Context(8) as ctx:
            for dist in (skel.COPY, skel.BLOCK):
                v = ctx.vector(x)
                v.set_distribution(dist)
                o = ctx.vector(n=n, dtype=np.int32)
                for _ in range(3):
                    ctx.scan(SUM_I32, v, o, np.int32(0))
                assert np.array_equal(o.download(), want), dist
            print("fallbacks", ctx.stats()["scan_coop_fallbacks"])
        print("OK")
    """)
    assert "OK" in out


def test_scan_next_to_an_sm_occupying_kernel():
    out = run("""
        SPIN = '''
        int spin(int x, long long cycles) {
            long long t0 = clock64();
            while (clock64() - t0 < cycles) { }
            return x;
        }'''
        n = (1 << 24) + 3
        x = si.uniform_int01(n, 78)
        want = oracle.skel_scan(SUM_I32, x, 0)
        hog = skel.Context(1)
        ctx = skel.Context(1)
        # enough spinning CTAs (one element each) to fill every SM for ~0.2 s
        h_in = hog.vector(np.zeros(148 * 2048 * 2, np.int32))
        h_out = hog.vector(n=h_in.n, dtype=np.int32)
        hog.map(SPIN, h_in, h_out, args=[np.int64(1000)])  # compile + warm
        hog.sync()
        v = ctx.vector(x)
        o = ctx.vector(n=n, dtype=np.int32)
        ctx.scan(SUM_I32, v, o, np.int32(0))  # compile + warm
        ctx.sync()
        for _ in range(3):
            hog.map(SPIN, h_in, h_out, args=[np.int64(20_000_000)])
            ctx.scan(SUM_I32, v, o, np.int32(0))
            assert np.array_equal(o.download(), want)
        hog.sync()
        ctx.close()
        hog.close()
        print("OK")
    """)
    assert "OK" in out
