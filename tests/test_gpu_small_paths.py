"""Reduce and Scan have two paths each: two short launches
for small vectors (tile aggregates, then a one-CTA fold / seeded tile scans),
the TMA kernels above SKEL_RED_SMALL_MAX / SKEL_SCAN_SMALL_MAX elements.  The
skeleton tests run at sizes that mostly take the small paths, so they are
re-run here in a subprocess with the switch points at 0 (everything through
the large-vector kernels) and at 10^9 (everything through the small paths) --
both stay under the same parity bars (eqs. (3), (4))."""
import os
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.mark.parametrize("small_max", ["0", "1000000000"])
def test_reduce_and_scan_tests_on_each_path(small_max):
    env = dict(os.environ, SKEL_SCAN_SMALL_MAX=small_max, SKEL_RED_SMALL_MAX=small_max)
    r = subprocess.run([sys.executable, "-m", "pytest", "-q", "-x", "-m", "gpu", "-k", "scan or reduce",
                        os.path.join(ROOT, "tests", "test_gpu_skeletons.py"),
                        os.path.join(ROOT, "tests", "test_gpu_distributions.py"),
                        os.path.join(ROOT, "tests", "test_gpu_graphs.py")],
                       env=env, capture_output=True, text=True, timeout=1200, cwd=ROOT)
    assert r.returncode == 0, r.stdout[-3000:] + r.stderr[-2000:]


def test_skeletons_without_programmatic_dependent_launches():
    """Every skeleton kernel is launched as a programmatic dependent of the
    previous kernel on its stream and waits (griddepcontrol.wait) before
    touching memory; with SKEL_PDL=0 the same kernels run with ordinary
    launches.  The skeleton, graph and distribution suites pass both ways."""
    env = dict(os.environ, SKEL_PDL="0")
    r = subprocess.run([sys.executable, "-m", "pytest", "-q", "-x", "-m", "gpu",
                        os.path.join(ROOT, "tests", "test_gpu_skeletons.py"),
                        os.path.join(ROOT, "tests", "test_gpu_graphs.py"),
                        os.path.join(ROOT, "tests", "test_gpu_distributions.py")],
                       env=env, capture_output=True, text=True, timeout=1500, cwd=ROOT)
    assert r.returncode == 0, r.stdout[-3000:] + r.stderr[-2000:]
