"""Vector buffers as VMM allocations (cuMemCreate + cuMemMap):
the skeleton, distribution and LM OSEM parity suites re-run with EVERY vector
buffer a VMM allocation (SKEL_VMM_MIN=0; by default buffers from 2 MB are), on
one device and on virtual devices -- the same bars as with cudaMalloc."""
import os
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def test_parity_suites_on_vmm_vectors():
    env = dict(os.environ, SKEL_VMM_MIN="0")
    r = subprocess.run([sys.executable, "-m", "pytest", "-q", "-x", "-m", "gpu",
                        os.path.join(ROOT, "tests", "test_gpu_skeletons.py"),
                        os.path.join(ROOT, "tests", "test_gpu_distributions.py"),
                        os.path.join(ROOT, "tests", "test_gpu_fused.py"),
                        os.path.join(ROOT, "tests", "test_gpu_coherence.py"),
                        os.path.join(ROOT, "tests", "test_gpu_lmosem.py"), "-k", "not full_size"],
                       env=env, capture_output=True, text=True, timeout=1800, cwd=ROOT)
    assert r.returncode == 0, r.stdout[-3000:] + r.stderr[-2000:]


def test_vmm_buffers_are_used():
    import numpy as np
    from paper_conf_ipps_steuwerkg11_b200 import skel
    with skel.Context(1) as ctx:
        v = ctx.vector(np.ones(1 << 22, np.float32))
        ctx.sync()
        assert ctx.stats()["vmm_allocs"] >= 1
        w = ctx.vector(n=1 << 22, dtype=np.float32)
        ctx.map("float f(float x){ return x + 1.0f; }", v, w)
        assert (w.download() == 2).all()
