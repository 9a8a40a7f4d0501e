"""World-size-2 CPU tests of the one-process-per-GPU (rank) path's host logic,
over torch.distributed with the gloo backend on 127.0.0.1.

The device exchanges of rank mode are NCCL collectives whose layouts are fixed
by the planner (parts of ceil(n/D), part k at offset k*ceil(n/D) of a full
buffer, padding to D*ceil(n/D)).  Here every rank builds exactly the buffers
the library would hold, runs the collective the planner names with gloo, and
the result must equal the oracle's distribution model.  The NCCL unique-id
bootstrap (rank 0 creates it, the others receive it) and the launch contract
of bench.py under torchrun are exercised too."""
import json
import os
import socket
import subprocess
import sys

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, n, q):
    sys.path.insert(0, ROOT)
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from oracle import distribution as odist
        from paper_conf_ipps_steuwerkg11_b200 import skel
        res = {}
        x = np.arange(n, dtype=np.float32) * 0.5 + 1
        lo, hi = skel.plan_part(n, world, rank)
        ps = -(-n // world)
        # block -> copy: in-place all-gather of padded parts
        assert skel.plan_exchange(skel.BLOCK, skel.COPY) == "allgather"
        part = torch.zeros(ps)
        part[: hi - lo] = torch.from_numpy(x[lo:hi])
        gathered = [torch.zeros(ps) for _ in range(world)]
        dist.all_gather(gathered, part)
        full = torch.cat(gathered)[:n].numpy()
        res["allgather"] = bool(np.array_equal(full, x))
        # copy -> block + add: reduce-scatter of D different copies (rank-dependent)
        assert skel.plan_exchange(skel.COPY, skel.BLOCK, skel.COMBINE_ADD) == "reduce_scatter"
        mine = np.zeros(ps * world, np.float32)
        mine[:n] = x * (rank + 1)
        t = torch.from_numpy(mine.copy())
        dist.all_reduce(t)  # gloo has no reduce_scatter: all-reduce, then keep part `rank` in place
        my_part = t.numpy()[rank * ps: rank * ps + (hi - lo)]
        copies = [x * (d + 1) for d in range(world)]
        model = odist.redistribute(copies, odist.COPY, odist.BLOCK, "add")
        res["reduce_scatter"] = bool(np.array_equal(my_part, model[rank]))
        # single -> block: scatter from rank 0 (root buffer padded to D*ceil(n/D))
        assert skel.plan_exchange(skel.SINGLE, skel.BLOCK) == "scatter"
        recv = torch.zeros(ps)
        if rank == 0:
            root = np.zeros(ps * world, np.float32)
            root[:n] = x
            dist.scatter(recv, [torch.from_numpy(root[k * ps:(k + 1) * ps].copy()) for k in range(world)], src=0)
        else:
            dist.scatter(recv, None, src=0)
        res["scatter"] = bool(np.array_equal(recv.numpy()[: hi - lo], odist.distribute(x, odist.BLOCK, world)[rank]))
        # cross-device Reduce: gather the D partials, fold in device order
        partial = torch.tensor([float(x[lo:hi].astype(np.float64).sum())], dtype=torch.float64)
        parts = [torch.zeros(1, dtype=torch.float64) for _ in range(world)]
        dist.all_gather(parts, partial)
        res["reduce"] = abs(sum(float(p) for p in parts) - float(x.astype(np.float64).sum())) < 1e-9
        # NCCL unique id: rank 0 creates, everyone receives the same 128 bytes
        obj = [skel.unique_id() if rank == 0 else None]
        dist.broadcast_object_list(obj, src=0)
        res["uid_len"] = len(obj[0])
        # without a GPU the rank context must fail loudly (no CPU fallback)
        if not torch.cuda.is_available():
            try:
                skel.Context(rank=rank, world=world, device=0, nccl_id=obj[0])
                res["no_fallback"] = False
            except skel.SkelError as e:
                res["no_fallback"] = e.name == "SKEL_ERR_CUDA"
        q.put((rank, res))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("n", [7, 1000, 6_300_000 // 100])
def test_rank_mode_exchanges_world2(n):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = free_port()
    procs = [ctx.Process(target=_worker, args=(r, 2, port, n, q)) for r in range(2)]
    for p in procs:
        p.start()
    out = dict(q.get(timeout=180) for _ in procs)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    for r in range(2):
        res = out[r]
        assert res["allgather"] and res["reduce_scatter"] and res["scatter"] and res["reduce"], res
        assert res["uid_len"] == 128
        assert res.get("no_fallback", True)


def test_bench_reference_arm_under_torchrun():
    """bench.py's launch contract at N = 2: rank 0 prints one JSON line, rank 1 exits 0."""
    port = free_port()
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node", "2",
           "--master-addr", "127.0.0.1", "--master-port", str(port), os.path.join(ROOT, "bench.py"),
           "--impl", "reference", "--gpus", "2", "--steps", "1", "--warmup", "3"]
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=600, cwd=ROOT)
    assert r.returncode == 0, r.stderr[-2000:]
    lines = [ln for ln in r.stdout.splitlines() if ln.startswith("{")]
    assert len(lines) == 1
    d = json.loads(lines[0])
    assert d["impl"] == "reference" and d["n_gpus"] == 2 and d["value"] > 0
    assert d["e2e"]["h2d_bytes_per_step"] == 0 and d["cpu_baseline"]["kind"] == "oracle"


def _cyclic_worker(rank, world, port, q):
    """Cyclic Mandelbrot rows at world 2 (mandelbrot.CyclicMandelbrot's layout):
    the permuted image is block-distributed with R = ceil(H/D) row slots per
    rank, slot t of rank k holding row k + t*D.  Each rank computes its slots
    with the oracle; gathered on rank 0 in block order and un-permuted (row r at
    slot (r mod D)*R + r div D) they must be the whole image, and the ranks'
    work (sum of counts) must be balanced."""
    sys.path.insert(0, ROOT)
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import oracle
        import skel_inputs as si
        from paper_conf_ipps_steuwerkg11_b200 import skel
        W, H, cap = 256, 190, 64   # H not a multiple of D: padding slots
        R = -(-H // world)
        n_perm = world * R * W
        lo, hi = skel.plan_part(n_perm, world, rank)
        assert (lo, hi) == (rank * R * W, (rank + 1) * R * W)
        pos = si.mandelbrot_positions(W, H).reshape(H, W)
        mine = np.zeros((R, W), np.int32)
        for t in range(R):
            row = rank + t * world
            if row < H:
                mine[t] = oracle.mandelbrot(np.ascontiguousarray(pos[row]), cap)
        parts = [torch.zeros(R * W, dtype=torch.int32) for _ in range(world)]
        dist.all_gather(parts, torch.from_numpy(mine.reshape(-1)))
        perm = torch.cat(parts).numpy().reshape(world * R, W)
        img = np.stack([perm[(r % world) * R + r // world] for r in range(H)])
        want = oracle.mandelbrot(np.ascontiguousarray(pos.reshape(-1)), cap).reshape(H, W)
        work = torch.tensor([float(mine.astype(np.int64).sum())], dtype=torch.float64)
        works = [torch.zeros(1, dtype=torch.float64) for _ in range(world)]
        dist.all_gather(works, work)
        w = np.array([float(x) for x in works])
        q.put((rank, {"image": bool(np.array_equal(img, want)), "balance": float(w.mean() / w.max())}))
    finally:
        dist.destroy_process_group()


def test_cyclic_rows_layout_world2():
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = free_port()
    procs = [ctx.Process(target=_cyclic_worker, args=(r, 2, port, q)) for r in range(2)]
    for p in procs:
        p.start()
    out = dict(q.get(timeout=180) for _ in procs)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    for r in range(2):
        assert out[r]["image"]
        assert out[r]["balance"] >= 0.95, out[r]
