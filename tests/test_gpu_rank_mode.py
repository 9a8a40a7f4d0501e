"""The one-process-per-GPU (rank) path of libskel, run with several processes
on the single available GPU.  Real NCCL refuses two ranks on one device, so
the ranks preload tests/fakenccl (a host-staged stand-in for the NCCL
collectives, test infrastructure): everything else -- buffer layouts, part
offsets, in-place collective conventions, cross-rank Reduce/Scan folds, LM
OSEM's all-gather / reduce-scatter, bench.py's torchrun path -- is the
product code."""
import json
import re
import os
import socket
import subprocess
import sys
from pathlib import Path

import pytest

pytestmark = pytest.mark.gpu
ROOT = Path(__file__).resolve().parents[1]


def free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


@pytest.fixture(scope="module")
def fake_nccl(tmp_path_factory):
    import nvidia.nccl as nn
    inc = Path(list(nn.__path__)[0]) / "include"
    out = tmp_path_factory.mktemp("fakenccl") / "libfakenccl.so"
    subprocess.run(["gcc", "-O2", "-shared", "-fPIC", "-I/usr/local/cuda/include", f"-I{inc}",
                    str(ROOT / "tests" / "fakenccl" / "fake_nccl.c"), "-o", str(out), "-L/usr/local/cuda/lib64",
                    "-lcudart", "-lpthread"], check=True, capture_output=True)
    return str(out)


def torchrun(nproc, script_args, fake, timeout=600, extra_env=None):
    # the host-staged fake collectives cannot be captured into CUDA graphs
    env = dict(os.environ, LD_PRELOAD=fake, SKEL_TEST_DEVICE="0", SKEL_BENCH_BACKEND="gloo", SKEL_BENCH_NO_GRAPH="1")
    env.update(extra_env or {})
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node", str(nproc),
           "--master-addr", "127.0.0.1", "--master-port", str(free_port()), *script_args]
    return subprocess.run(cmd, capture_output=True, text=True, timeout=timeout, cwd=str(ROOT), env=env)


@pytest.mark.parametrize("nproc", [2, 3])
def test_rank_mode_selftest(fake_nccl, nproc):
    r = torchrun(nproc, ["tools/rank_selftest.py"], fake_nccl)
    assert r.returncode == 0, r.stdout[-3000:] + r.stderr[-3000:]
    # one "rank k/n device d: OK" report per rank (the ranks' lines may interleave)
    oks = re.findall(r"rank (\d+)/\d+ device \d+: OK", r.stdout)
    assert sorted(map(int, oks)) == list(range(nproc)), r.stdout[-2000:]


def test_bench_rank_path(fake_nccl):
    r = torchrun(2, ["bench.py", "--gpus", "2", "--steps", "3", "--warmup", "3", "--log2n", "22", "--e2e-steps", "1",
                     "--no-cpu"], fake_nccl)
    assert r.returncode == 0, r.stdout[-3000:] + r.stderr[-3000:]
    lines = [ln for ln in r.stdout.splitlines() if ln.startswith("{")]
    assert len(lines) == 1
    d = json.loads(lines[0])
    assert d["n_gpus"] == 2 and d["value"] > 0 and d["config"]["distribution"] == "block"
    assert d["e2e"]["h2d_bytes_per_step"] == 2 * (1 << 22) * 4  # this rank's parts of x and y
    assert d["mandelbrot"]["sum_iter"] == 453197644
    assert d["mandelbrot"]["all_bit_identical"] and d["mandelbrot"]["cap4096"]["sum_iter"] > 453197644
    ex = d["lmosem"]["exchange"]  # reduce-scatter / all-gather of the 25.2 MB image alone
    assert ex["bytes"] == 150 * 150 * 280 * 4 and ex["reduce_scatter_busbw_GBps"] > 0 and ex["all_gather_busbw_GBps"] > 0
    assert d["lmosem"]["full_recon_s"] > 0


def test_rank_mode_nccl_windows_fall_back(fake_nccl):
    """SKEL_NCCL_WINDOWS=1: the fused LM OSEM tail asks NCCL for symmetric
    windows (ncclMemAlloc + ncclCommWindowRegister).  The
    host-staged stand-in has no such memory, so every rank must agree to fall
    back to CUDA IPC -- the self-test (incl. the fused tail against the oracle)
    still passes at 2 ranks."""
    r = torchrun(2, ["tools/rank_selftest.py"], fake_nccl, extra_env={"SKEL_NCCL_WINDOWS": "1"})
    assert r.returncode == 0, r.stdout[-3000:] + r.stderr[-3000:]
    oks = re.findall(r"rank (\d+)/\d+ device \d+: OK", r.stdout)
    assert sorted(map(int, oks)) == [0, 1], r.stdout[-2000:]


def real_nccl_run(nproc, script_args, timeout=300, extra_env=None):
    """torchrun WITHOUT the stand-in: the ranks load the real NCCL (the one
    libskel links).  One GPU, so one rank: NCCL refuses two ranks on a device."""
    env = dict(os.environ, SKEL_TEST_DEVICE="0", SKEL_BENCH_BACKEND="gloo")
    env.pop("LD_PRELOAD", None)
    env.update(extra_env or {})
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node", str(nproc),
           "--master-addr", "127.0.0.1", "--master-port", str(free_port()), *script_args]
    return subprocess.run(cmd, capture_output=True, text=True, timeout=timeout, cwd=str(ROOT), env=env)


@pytest.mark.parametrize("windows", ["0", "1"])
def test_rank_mode_real_nccl_one_rank(windows):
    """The rank path on the REAL NCCL library with a one-rank communicator
    (ncclCommInitRank): the self-test's skeletons and transitions, and LM OSEM's
    fused tail forced onto the rank path (SKEL_FORCE_MULTIMEM=1) -- its
    ncclAllGather of the CUDA IPC handles and ncclAllReduce barriers, or with
    SKEL_NCCL_WINDOWS=1 ncclMemAlloc + ncclCommWindowRegister(
    NCCL_WIN_COLL_SYMMETRIC) + ncclDevCommCreate for the tail's vectors (or the
    ranks' agreed fallback when NCCL declines) -- checked against the oracle."""
    # SKEL_FORCE_MULTIMEM=1: a one-rank communicator takes the fused tail too
    r = real_nccl_run(1, ["tools/rank_selftest.py"],
                      extra_env={"SKEL_NCCL_WINDOWS": windows, "SKEL_LOG": "1", "SKEL_FORCE_MULTIMEM": "1"})
    assert r.returncode == 0, r.stdout[-3000:] + r.stderr[-3000:]
    assert re.search(r"rank 0/1 device \d+: OK", r.stdout), r.stdout[-2000:] + r.stderr[-2000:]
    if windows == "1":  # the outcome of the window set-up is logged either way
        assert "NCCL symmetric window" in r.stderr, r.stderr[-2000:]
        print([ln for ln in r.stderr.splitlines() if "NCCL symmetric window" in ln][:2])
