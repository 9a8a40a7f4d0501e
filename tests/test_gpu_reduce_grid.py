"""Reduce grid policy: the oversubscribed grid (several CTAs
per resident slot, contiguous tile ranges, last-CTA ordered fold over more
partials) must keep index order for non-commutative operators.

The policy only oversubscribes above ~55 tiles per SM, so (a) a subprocess
forces it at small, ragged sizes through the SKEL_RED_OVERSUB tuning hook
(read once per process), and (b) one case runs at a size where the default
policy oversubscribes by itself (2^26 16-byte elements, 1 GiB).  Both compare
bit for bit with the oracle's left fold (eq. (3))."""
import os
import subprocess
import sys
import textwrap

import numpy as np
import pytest

import oracle
from paper_conf_ipps_steuwerkg11_b200 import skel

from test_gpu_skeletons import AFF, AFF2, AFF3, A2, M2, MAT_U, rand_struct

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))

CHILD = textwrap.dedent("""
    import sys
    sys.path[:0] = [{root!r}, {tests!r}]
    import numpy as np
    import oracle
    import skel_inputs as si
    from paper_conf_ipps_steuwerkg11_b200 import skel
    from paper_conf_ipps_steuwerkg11_b200.workloads import SUM_F32, SUM_I32
    from test_gpu_skeletons import AFF, AFF2, AFF3, A2, M2, MAT_U, rand_struct
    bad = []
    with skel.Context(1) as ctx:
        for n in (1, 4095, 4097, 3 * 4096 + 5, 100_003, 1_000_001):
            m = rand_struct(M2, n, n)
            if ctx.reduce(MAT_U, ctx.vector(m)).tobytes() != oracle.skel_reduce(MAT_U, m).tobytes():
                bad.append(("M2", n))
        for n in (8191, 8193, 500_001):
            m = rand_struct(A2, n, n + 1)
            if ctx.reduce(AFF2, ctx.vector(m)).tobytes() != oracle.skel_reduce(AFF2, m).tobytes():
                bad.append(("A2", n))
            a = rand_struct(AFF, n, n + 2)
            if ctx.reduce(AFF3, ctx.vector(a)).tobytes() != oracle.skel_reduce(AFF3, a).tobytes():
                bad.append(("AFF3", n))
        for n in (16383, 16385, 2_000_003):
            x = si.uniform_int01(n, 7)
            if int(ctx.reduce(SUM_I32, ctx.vector(x))) != int(x.astype(np.int64).sum()):
                bad.append(("i32", n))
            xf = si.uniform_f32(n, 8)
            r = float(ctx.reduce(SUM_F32, ctx.vector(xf)))
            if abs(r - oracle.sum_f32_exact(xf)) > 1e-5 * oracle.abssum_f32(xf):
                bad.append(("f32", n))
    print("BAD", bad)
    sys.exit(1 if bad else 0)
""")


@pytest.mark.parametrize("oversub", ["3", "8"])
def test_forced_oversubscription_keeps_order(oversub):
    env = dict(os.environ, SKEL_RED_OVERSUB=oversub)
    code = CHILD.format(root=ROOT, tests=os.path.join(ROOT, "tests"))
    r = subprocess.run([sys.executable, "-c", code], env=env, capture_output=True, text=True, timeout=900)
    assert r.returncode == 0, r.stdout[-2000:] + r.stderr[-2000:]


def test_default_policy_oversubscribes_large_noncommutative():
    n = 1 << 26  # 16-byte elements: 16384 tiles of 64 KB -> 2 CTAs per slot
    m = rand_struct(M2, n, 2026)
    with skel.Context(1) as ctx:
        got = ctx.reduce(MAT_U, ctx.vector(m))
    assert got.tobytes() == oracle.skel_reduce(MAT_U, m).tobytes()
