#!/usr/bin/env python3
"""Benchmark of the SkelCL hot path on B200 (BASELINE.json configs).

Headline (BASELINE.json configs[1]): one *step* = Map(x*2+1) + Zip(saxpy) +
Reduce(+) + Scan(+) over float32 vectors of 2^30 elements per GPU (4 GiB each,
far larger than the 126 MB L2, so no flush is needed), through libskel's
C-ABI.  value = aggregate algorithmic GB/s of the step over all GPUs
(32 bytes/element: Map 8, Zip 12, Reduce 4, Scan 8).  Side measurements in
the same run: per-skeleton GB/s and %HBM, Mandelbrot 4096x3072 (configs[2],
Mpix/s) and one LM OSEM subset of 10^6 events (configs[3]/[4], seconds).

    python bench.py [--gpus N] [--steps K] [--warmup W] [--impl skel|reference]
    torchrun --nproc-per-node N bench.py --gpus N ...   (one process per GPU)

`--impl reference` times the CPU oracle (the task's reference arm) on host
cores for the same metric on a bounded sample.
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import threading
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

BYTES_PER_ELEM = {"map": 8, "zip": 12, "reduce": 4, "scan": 8}
STEP_BYTES = sum(BYTES_PER_ELEM.values())
METRIC = "skeleton step GB/s (Map+Zip+Reduce+Scan, float32, 2^30 elements per GPU)"
SEED = 20110516


# untimed launches of a skeleton before it is timed: its first launch compiles
# (or loads) the module and decides the element-wise grid policy on a sample
# (runtime.cpp ew_decide; no trial policies on user launches)
TUNE = 1


def bench_config(nloc: int, world: int) -> dict:
    """The workload description shared by the GPU arm and the reference arm."""
    return {"workload": "configs[1]: Reduce(+)/Zip(saxpy)/Scan(+) (+ Map x*2+1) sweep point "
                        "n=2^30 float32 per GPU, one step = all four skeletons",
            "elements_per_gpu": nloc, "elements_total": nloc * world,
            "distribution": "single" if world == 1 else "block",
            "l2": "inputs (4 GiB per vector) far exceed the 126 MB L2; no flush needed"}


def env_world():
    return int(os.environ.get("WORLD_SIZE", "1")), int(os.environ.get("RANK", "0")), \
        int(os.environ.get("LOCAL_RANK", "0"))


def measured_peaks():
    p = os.path.join(ROOT, "MEASURED_PEAKS.json")
    try:
        with open(p) as fh:
            d = json.load(fh)
        return float(d["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs)"
    except Exception:
        return 6650.0, "fallback (B200_PROFILING.md: 6.65 TB/s)"


def traffic_table():
    p = os.path.join(ROOT, "profiles", "traffic.json")
    try:
        with open(p) as fh:
            return json.load(fh)
    except Exception:
        return {}


class ClockSampler:
    """nvidia-smi clocks + throttle reasons sampled during the timed region."""

    FIELDS = ("index,clocks.sm,clocks.max.sm,power.draw,clocks_event_reasons.active,"
              "clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
              "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap")

    def __init__(self, gpu: int):
        self.gpu = gpu
        self.proc = None
        self.lines = []

    def start(self):
        try:
            self.proc = subprocess.Popen(["nvidia-smi", "-i", str(self.gpu), f"--query-gpu={self.FIELDS}",
                                          "--format=csv,noheader,nounits", "-lms", "100"],
                                         stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
            self.t = threading.Thread(target=self._read, daemon=True)
            self.t.start()
        except Exception:
            self.proc = None

    def _read(self):
        for line in self.proc.stdout:
            self.lines.append(line.strip())

    def stop(self):
        if not self.proc:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["nvidia-smi unavailable"]}
        time.sleep(0.25)
        self.proc.terminate()
        try:
            self.proc.wait(timeout=5)
        except Exception:
            self.proc.kill()
        sm, smax, reasons = [], None, set()
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        for ln in self.lines:
            f = [x.strip() for x in ln.split(",")]
            if len(f) < 9:
                continue
            try:
                sm.append(float(f[1]))
                smax = float(f[2])
            except ValueError:
                continue
            for nm, val in zip(names, f[5:9]):
                if val.lower().startswith("active"):
                    reasons.add(nm)
        return {"sm_mhz": statistics.median(sm) if sm else None, "sm_max_mhz": smax,
                "reasons": sorted(reasons), "samples": len(sm)}


# ---------------------------------------------------------------------------
# CPU oracle timing (cpu_baseline and the --impl reference arm)
# ---------------------------------------------------------------------------
def oracle_step(x, y):
    import oracle
    from paper_conf_ipps_steuwerkg11_b200.workloads import MAP_F32, SAXPY_F32
    oracle.skel_map(MAP_F32, x, np.float32)
    oracle.skel_zip(SAXPY_F32, x, y, np.float32, args=[np.float32(2.5)])
    oracle.sum_f32_exact(x)
    oracle.exscan_f32_exact(x)


def cpu_baseline(total_log2=30, chunk_log2=26):
    """The oracle as it stands (single-threaded C), timed on this host on a
    bounded sample: 2^total elements processed in chunks of 2^chunk."""
    import skel_inputs as si
    chunks = 1 << (total_log2 - chunk_log2)
    n = 1 << chunk_log2
    oracle_step(si.uniform_f32(1024, 1), si.uniform_f32(1024, 2))  # compile the user functions
    t = 0.0
    for c in range(chunks):
        x, y = si.uniform_f32(n, SEED + 2 * c), si.uniform_f32(n, SEED + 2 * c + 1)
        t0 = time.perf_counter()
        oracle_step(x, y)
        t += time.perf_counter() - t0
    elems = chunks * n
    return {"value": STEP_BYTES * elems / t / 1e9, "unit": "GB/s", "cores": 1, "kind": "oracle",
            "sample": f"Map+Zip+Reduce+Scan oracle over 2^{total_log2} float32 elements "
                      f"({chunks} chunks of 2^{chunk_log2}), {t:.1f} s single-threaded",
            "host_cpus": os.cpu_count()}


def host_info() -> dict:
    """The host the oracle runs on: logical CPUs, the ones this process may
    use, and lscpu's model name."""
    model = None
    try:
        out = subprocess.run(["lscpu"], capture_output=True, text=True, timeout=10).stdout
        for ln in out.splitlines():
            if ln.lower().startswith("model name"):
                model = ln.split(":", 1)[1].strip()
                break
    except Exception:
        pass
    try:
        usable = len(os.sched_getaffinity(0))
    except Exception:
        usable = os.cpu_count()
    return {"host_cpus": os.cpu_count(), "usable_cpus": usable, "cpu_model": model}


def _threads() -> int:
    return max(1, host_info()["usable_cpus"] or 1)


def _par(fn, items, threads):
    """Run fn over items on `threads` host threads (the oracle's C loops release
    the GIL, so disjoint chunks run side by side)."""
    from concurrent.futures import ThreadPoolExecutor
    if threads <= 1:
        return [fn(it) for it in items]
    with ThreadPoolExecutor(max_workers=threads) as ex:
        return list(ex.map(fn, items))


def oracle_step_allcores(x, y, threads):
    """oracle_step on all host cores: Map/Zip/Reduce on disjoint chunks; Scan as
    chunk sums (float64) then seeded chunk scans (oracle_exscan_f32_seeded)."""
    import oracle
    from paper_conf_ipps_steuwerkg11_b200.workloads import MAP_F32, SAXPY_F32
    n = x.size
    cuts = np.linspace(0, n, threads + 1).astype(np.int64)
    rng = list(zip(cuts[:-1], cuts[1:]))
    m, z, s = np.empty_like(x), np.empty_like(x), np.empty_like(x)

    def mz(r):
        a, b = r
        m[a:b] = oracle.skel_map(MAP_F32, x[a:b], np.float32)
        z[a:b] = oracle.skel_zip(SAXPY_F32, x[a:b], y[a:b], np.float32, args=[np.float32(2.5)])
    _par(mz, rng, threads)
    sums = _par(lambda r: oracle.sum_f32_exact(x[r[0]:r[1]]), rng, threads)
    pre = np.concatenate([[0.0], np.cumsum(sums)])
    _par(lambda k: oracle.exscan_f32_seeded(x[rng[k][0]:rng[k][1]], pre[k], s[rng[k][0]:rng[k][1]]),
         range(len(rng)), threads)
    return float(pre[-1])


def cpu_baseline_allcores(total_log2=30, chunk_log2=26):
    """The skeleton step's oracle on every usable host core (same bounded sample
    as cpu_baseline)."""
    import skel_inputs as si
    T = _threads()
    chunks = 1 << (total_log2 - chunk_log2)
    n = 1 << chunk_log2
    oracle_step(si.uniform_f32(1024, 1), si.uniform_f32(1024, 2))
    t = 0.0
    for c in range(chunks):
        x, y = si.uniform_f32(n, SEED + 2 * c), si.uniform_f32(n, SEED + 2 * c + 1)
        t0 = time.perf_counter()
        oracle_step_allcores(x, y, T)
        t += time.perf_counter() - t0
    return {"value": STEP_BYTES * chunks * n / t / 1e9, "unit": "GB/s", "cores": T, "kind": "oracle (all cores)",
            "sample": f"the same 2^{total_log2} elements in {chunks} chunks of 2^{chunk_log2}, each split over {T} "
                      f"threads (scan: chunk sums, then seeded chunk scans), {t:.1f} s"}


def cpu_baseline_mandelbrot():
    """Oracle (eq. (5), oracle_mandelbrot) for configs[0] and configs[2]: one
    thread, and every usable core over row bands."""
    import oracle
    import skel_inputs as si
    T = _threads()
    res = {}
    for tag, (w, h) in (("configs0_1024x768", (1024, 768)), ("configs2_4096x3072", (4096, 3072))):
        pos = si.mandelbrot_positions(w, h)
        t0 = time.perf_counter()
        oracle.mandelbrot(pos, 256)
        t1 = time.perf_counter() - t0
        cuts = np.linspace(0, pos.size, 4 * T + 1).astype(np.int64)
        t0 = time.perf_counter()
        _par(lambda k: oracle.mandelbrot(pos[cuts[k]:cuts[k + 1]], 256), range(4 * T), T)
        tT = time.perf_counter() - t0
        res[tag] = {"ms_1core": t1 * 1e3, "Mpix_per_s_1core": pos.size / t1 / 1e6,
                    "ms_allcores": tT * 1e3, "Mpix_per_s_allcores": pos.size / tT / 1e6}
    return {"kind": "oracle", "unit": "Mpix/s", "cores": T, "value": res["configs2_4096x3072"]["Mpix_per_s_1core"],
            "sample": "whole images, cap 256 (value: configs[2] on 1 core)", **res}


def _lm_allcores(ev, f, T):
    """Listing 3 for one subset on T threads: each thread's chunk of events
    into a private error image (oracle_lmosem_error_image), the images summed,
    then the update (oracle_lmosem_update)."""
    import oracle
    cuts = np.linspace(0, ev.size, T + 1).astype(np.int64)
    parts = _par(lambda k: oracle.lmosem_error_image(ev[cuts[k]:cuts[k + 1]], f)[0], range(T), T)
    c = parts[0]
    for p in parts[1:]:
        c += p
    return oracle.lmosem_update(f, c)


def cpu_baseline_lmosem(subsets):
    """Oracle LM OSEM (Listing 3): one subset on one core, the same subset and
    the full 10-subset reconstruction (configs[4], once per job) on all cores."""
    import oracle
    T = _threads()
    nvox = 150 * 150 * 280
    f0 = np.ones(nvox, np.float64)
    t0 = time.perf_counter()
    oracle.lmosem_subset(subsets[0], f0)
    t1 = time.perf_counter() - t0
    t0 = time.perf_counter()
    _lm_allcores(subsets[0], f0, T)
    tT = time.perf_counter() - t0
    t0 = time.perf_counter()
    f = f0.copy()
    for ev in subsets:
        f = _lm_allcores(ev, f, T)
    tR = time.perf_counter() - t0
    return {"kind": "oracle", "unit": "s", "cores": T, "value": t1,
            "sample": f"one subset of {subsets[0].size} events on 1 core (value), on {T} cores, and the "
                      f"{len(subsets)}-subset reconstruction on {T} cores",
            "subset_s_1core": t1, "subset_s_allcores": tT, "full_recon_s_allcores": tR}


def run_reference(args):
    world, rank, _ = env_world()
    if rank != 0:
        return
    import skel_inputs as si
    n = 1 << 24
    x, y = si.uniform_f32(n, SEED), si.uniform_f32(n, SEED + 1)
    for _ in range(args.warmup):
        oracle_step(x, y)
    t0 = time.perf_counter()
    for _ in range(args.steps):
        oracle_step(x, y)
    dt = (time.perf_counter() - t0) / args.steps
    value = STEP_BYTES * n / dt / 1e9
    line = {"impl": "reference", "metric": METRIC, "value": value, "unit": "GB/s", "n_gpus": args.gpus,
            "steps": args.steps, "warmup": args.warmup, "ms_per_step": dt * 1e3, "higher_is_better": True,
            "scaling": "weak", "vs_baseline": None, "dtype": "f32", "data": "synthetic",
            "config": bench_config(1 << args.log2n, args.gpus),
            "cpu_baseline": {"value": value, "unit": "GB/s", "cores": 1, "kind": "oracle",
                             "sample": f"bounded: each step runs the oracle on 2^24 of the 2^30 float32 elements "
                                       f"({args.steps} steps, single-threaded C); value scaled per byte"},
            "e2e": {"value": value, "unit": "GB/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)


# ---------------------------------------------------------------------------
# GPU arm
# ---------------------------------------------------------------------------
def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=20)
    ap.add_argument("--warmup", type=int, default=5)
    ap.add_argument("--impl", default="skel", choices=["skel", "reference"])
    ap.add_argument("--log2n", type=int, default=30, help="elements per GPU (log2)")
    ap.add_argument("--e2e-steps", type=int, default=8)
    ap.add_argument("--no-extras", action="store_true", help="skip Mandelbrot / LM OSEM side measurements")
    ap.add_argument("--no-cpu", action="store_true", help="skip the cpu_baseline oracle timing")
    args = ap.parse_args()
    args.warmup = max(args.warmup, 3)

    if args.impl == "reference":
        run_reference(args)
        return

    import torch
    import torch.distributed as dist

    from paper_conf_ipps_steuwerkg11_b200 import skel
    from paper_conf_ipps_steuwerkg11_b200.workloads import MAP_F32, SAXPY_F32, SUM_F32

    world, rank, local = env_world()
    # test hooks: SKEL_TEST_DEVICE puts every rank on one device (rank-mode tests on a
    # single GPU with tests/fakenccl), SKEL_BENCH_BACKEND=gloo for the process group
    local = int(os.environ.get("SKEL_TEST_DEVICE", local))
    backend = os.environ.get("SKEL_BENCH_BACKEND", "nccl")
    torch.cuda.set_device(local)
    if world > 1:
        if backend == "nccl":
            dist.init_process_group("nccl", device_id=torch.device("cuda", local))
        else:
            dist.init_process_group(backend)
        obj = [skel.unique_id() if rank == 0 else None]
        dist.broadcast_object_list(obj, src=0)
        ctx = skel.Context(rank=rank, world=world, device=local, nccl_id=obj[0])
    else:
        ctx = skel.Context(1)

    def barrier():
        if world > 1:
            dist.barrier()

    def max_over_ranks(v: float) -> float:
        if world == 1:
            return v
        t = torch.tensor([v], device="cuda" if backend == "nccl" else "cpu", dtype=torch.float64)
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
        return float(t.item())

    stream = torch.cuda.ExternalStream(ctx.stream(0), device=torch.device("cuda", local))
    nloc = 1 << args.log2n
    N = nloc * world
    import skel_inputs as si

    # ---- inputs: this rank's block of x, y (uniform [0,1), PCG64), uploaded once
    x = ctx.vector(n=N, dtype=np.float32)
    y = ctx.vector(n=N, dtype=np.float32)
    lo = rank * nloc
    if world > 1:
        x.set_distribution(skel.BLOCK)
        y.set_distribution(skel.BLOCK)
    x.upload_part(lo, si.uniform_f32(nloc, SEED + 2 * rank))
    y.upload_part(lo, si.uniform_f32(nloc, SEED + 2 * rank + 1))
    m = ctx.vector(n=N, dtype=np.float32)
    z = ctx.vector(n=N, dtype=np.float32)
    s = ctx.vector(n=N, dtype=np.float32)
    r = ctx.vector(n=1, dtype=np.float32)
    a = np.float32(2.5)
    for kind, src in (("map", MAP_F32), ("zip", SAXPY_F32), ("reduce", SUM_F32)):
        ctx.prepare(kind, src)

    def step(ev=None):
        if ev is not None:
            ev[0].record(stream)
        ctx.map(MAP_F32, x, m)
        if ev is not None:
            ev[1].record(stream)
        ctx.zip(SAXPY_F32, x, y, z, args=[a])
        if ev is not None:
            ev[2].record(stream)
        ctx.reduce_to(SUM_F32, x, r)
        if ev is not None:
            ev[3].record(stream)
        ctx.scan(SUM_F32, x, s, np.float32(0))
        if ev is not None:
            ev[4].record(stream)

    for _ in range(TUNE + args.warmup):  # grid-policy trials first, then the warm-up proper
        step()
    ctx.sync()

    evs = [[torch.cuda.Event(enable_timing=True) for _ in range(5)] for _ in range(args.steps)]
    t_start, t_stop = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    sampler = ClockSampler(local)
    launches0 = ctx.stats()["kernel_launches"]
    xfer0 = ctx.stats()
    barrier()
    torch.cuda.synchronize()
    sampler.start()
    time.sleep(0.3)
    torch.cuda.nvtx.range_push("timed")  # ncu --nvtx --nvtx-include timed/ selects the timed launches
    t_start.record(stream)
    for k in range(args.steps):
        step(evs[k])
    t_stop.record(stream)
    torch.cuda.nvtx.range_pop()
    ctx.sync()
    torch.cuda.synchronize()
    barrier()
    clocks = sampler.stop()
    st1 = ctx.stats()
    launches = st1["kernel_launches"] - launches0
    assert st1["h2d_bytes"] == xfer0["h2d_bytes"], "inputs were not resident in the timed region"
    ms_total = max_over_ranks(t_start.elapsed_time(t_stop))
    ms_step = ms_total / args.steps
    per = {}
    for i, name in enumerate(("map", "zip", "reduce", "scan")):
        ts = [evs[k][i].elapsed_time(evs[k][i + 1]) for k in range(args.steps)]
        avg = max_over_ranks(sum(ts) / len(ts))
        per[name] = {"ms": avg, "GBps": BYTES_PER_ELEM[name] * nloc / (avg * 1e-3) / 1e9}
    value = STEP_BYTES * N / (ms_step * 1e-3) / 1e9
    peak, peak_src = measured_peaks()
    for name in per:
        per[name]["frac_of_hbm"] = per[name]["GBps"] / peak
    dom = max(per, key=lambda k: per[k]["ms"])
    traffic = traffic_table().get(dom)
    roofline = {"bound": "hbm", "kernel": dom, "achieved": per[dom]["GBps"], "peak": peak, "unit": "GB/s",
                "frac": per[dom]["GBps"] / peak, "peak_source": peak_src,
                "algorithmic_bytes_per_launch": BYTES_PER_ELEM[dom] * nloc,
                "traffic": traffic, "traffic_source": "profiles/traffic.json (ncu --set full)" if traffic else None}

    # ---- end to end through the C-ABI: pinned host inputs -> every result on the host
    e2e = None
    if args.e2e_steps > 0:
        # the user's result buffers (pinned host memory)
        hbufs = [torch.empty(nloc, dtype=torch.float32, pin_memory=True).numpy() for _ in range(3)]
        ctx.sync()
        barrier()
        st0 = ctx.stats()
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        for _ in range(args.e2e_steps):
            x.mark_host_modified()
            y.mark_host_modified()
            ctx.map(MAP_F32, x, m)
            ctx.zip(SAXPY_F32, x, y, z, args=[a])
            ctx.scan(SUM_F32, x, s, np.float32(0))
            ctx.reduce(SUM_F32, x)  # blocking: the scalar on the host
            # this rank's block of every output vector to the host, asynchronously:
            # the copies overlap the next step's uploads (opposite PCIe direction)
            for v, hb in zip((m, z, s), hbufs):
                v.download_part_async(lo, hb)
        ctx.sync()  # every download has landed
        dt = max_over_ranks(time.perf_counter() - t0) / args.e2e_steps
        st1 = ctx.stats()
        e2e = {"value": STEP_BYTES * N / dt / 1e9, "unit": "GB/s", "ms_per_step": dt * 1e3,
               "h2d_bytes_per_step": (st1["h2d_bytes"] - st0["h2d_bytes"]) // args.e2e_steps,
               "d2h_bytes_per_step": (st1["d2h_bytes"] - st0["d2h_bytes"]) // args.e2e_steps,
               "path": "skel_vector_mark_host_modified on pinned host mirrors of x, y, then map/zip/scan/reduce "
                       "(lazy H2D inside), skel_reduce's blocking D2H of the scalar, and "
                       "skel_vector_download_part_async of the Map, Zip and Scan outputs into pinned host buffers "
                       "(overlapping the next step's uploads); skel_sync after the last step"}
        del hbufs

    # free the big vectors before the side measurements
    for v in (x, y, m, z, s):
        v.destroy()

    extras = {}
    if not args.no_extras:
        extras["sweep"] = bench_sweep(ctx, skel, stream, world, rank, barrier, max_over_ranks, args)
        if world == 1:
            extras["overhead"] = bench_overhead(ctx, skel, stream, args)
        extras["mandelbrot"] = bench_mandelbrot(ctx, skel, stream, world, rank, barrier, max_over_ranks, args)
        extras["lmosem"] = bench_lmosem(ctx, skel, stream, world, rank, barrier, max_over_ranks, args)

    cpu = None
    if rank == 0 and world == 1 and not args.no_cpu:
        cpu = cpu_baseline()
        cpu.update(host_info())
        cpu["allcores"] = cpu_baseline_allcores()
        if "mandelbrot" in extras:
            extras["mandelbrot"]["cpu_baseline"] = cpu_baseline_mandelbrot()
        if "lmosem" in extras:
            extras["lmosem"]["cpu_baseline"] = cpu_baseline_lmosem(lm_subsets(1_000_000, 10, 0, 1_000_000))

    if rank == 0:
        line = {"metric": METRIC, "value": value, "unit": "GB/s", "n_gpus": world, "steps": args.steps,
                "warmup": args.warmup, "ms_per_step": ms_step, "higher_is_better": True, "scaling": "weak",
                "vs_baseline": None, "dtype": "f32", "data": "synthetic (PCG64 uniform [0,1) float32)",
                "config": bench_config(nloc, world),
                "per_skeleton": per, "roofline": roofline, "cpu_baseline": cpu, "e2e": e2e,
                "gpu_launches": launches, "clocks": clocks, **extras}
        print(json.dumps(line), flush=True)
    ctx.close()
    if world > 1:
        dist.destroy_process_group()


def bench_sweep(ctx, skel, stream, world, rank, barrier, max_over_ranks, args):
    """configs[1] sweep: GB/s per skeleton, n = 2^20 .. 2^30 per GPU, float32 and int32.
    Vectors are filled on the device (values do not change the memory traffic).
    Sizes whose operands fit in 4x L2 rotate over R independent operand sets
    (R x footprint >= 4x L2, R >= 2): one timed repetition is a CUDA graph of R
    back-to-back launches, each on a set last touched R launches earlier, so
    every launch starts with its operands evicted from L2 and the graph launch
    overhead is amortised (steady-state throughput, not one-launch latency)."""
    import math

    import torch
    from paper_conf_ipps_steuwerkg11_b200.workloads import (MAP_F32, MAP_I32, SAXPY_F32, SAXPY_I32, SUM_F32,
                                                             SUM_I32)
    funcs = {np.float32: (MAP_F32, SAXPY_F32, SUM_F32), np.int32: (MAP_I32, SAXPY_I32, SUM_I32)}
    peak, _ = measured_peaks()
    l2 = 126e6
    out = []
    for dt, (fm, fz, fs) in funcs.items():
        for k in range(20, 31, 2):
            nloc = 1 << k
            N = nloc * world
            small = 3 * nloc * 4 < 4 * l2
            R = max(2, min(64, math.ceil(4 * l2 / (3 * nloc * 4)))) if small else 1
            sets = []
            for _ in range(R):
                x, y, o = (ctx.vector(n=N, dtype=dt) for _ in range(3))
                r = ctx.vector(n=1, dtype=dt)
                for v, val in ((x, 1), (y, 2)):
                    if world > 1:
                        v.fill_dist(skel.BLOCK, dt(val))
                    else:
                        v.fill(dt(val))
                sets.append((x, y, o, r))
            a = dt(3)
            ops = {"map": lambda st: ctx.map(fm, st[0], st[2]),
                   "zip": lambda st: ctx.zip(fz, st[0], st[1], st[2], args=[a]),
                   "reduce": lambda st: ctx.reduce_to(fs, st[0], st[3]),
                   "scan": lambda st: ctx.scan(fs, st[0], st[2], dt(0))}
            reps = 10 if k < 30 else 5
            row = {"dtype": np.dtype(dt).name, "log2n": k,
                   "l2": f"rotating {R} operand sets (>= 4x L2)" if small else "exceeds L2"}
            for name, op in ops.items():
                def fn(op=op):
                    for st in sets:
                        op(st)
                for _ in range(2):
                    fn()
                ctx.sync()
                try:  # replay as a CUDA graph: no host overhead in the timing
                    if os.environ.get("SKEL_BENCH_NO_GRAPH"):
                        raise skel.SkelError(8, "graphs disabled")
                    g = ctx.capture(fn)
                    g.launch()
                    ctx.sync()
                    run = g.launch
                except skel.SkelError:  # e.g. a collective backend that cannot be captured
                    g, run = None, fn
                    row["graph"] = False
                barrier()
                torch.cuda.synchronize()
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                e0.record(stream)
                for _ in range(reps):
                    run()
                e1.record(stream)
                ctx.sync()
                if g is not None:
                    g.destroy()
                ms = max_over_ranks(e0.elapsed_time(e1) / (reps * R))
                gbs = BYTES_PER_ELEM[name] * N / (ms * 1e-3) / 1e9
                row[name] = {"ms": round(ms, 5), "GBps": round(gbs, 1), "frac": round(gbs / world / peak, 4)}
            out.append(row)
            for st in sets:
                for v in st:
                    v.destroy()
    return out


def bench_overhead(ctx, skel, stream, args):
    """NEXT-3: (a) the skeletons vs the same operations hand-written in CUDA C++
    (nvcc, float4 loops) and CUB's DeviceScan, on the same device buffers and
    stream -- the analog of the paper's SkelCL-vs-OpenCL overhead;
    (b) NVRTC build time vs loading the cubin from the disk cache."""
    import ctypes
    import tempfile
    import torch
    from paper_conf_ipps_steuwerkg11_b200.workloads import MAP_F32, SAXPY_F32, SUM_F32
    hw = ctypes.CDLL(os.path.join(ROOT, "paper_conf_ipps_steuwerkg11_b200", "libhandwritten.so"))
    P, S = ctypes.c_void_p, ctypes.c_size_t
    hw.hw_map_f32.argtypes = [P, P, S, P]
    hw.hw_saxpy_f32.argtypes = [P, P, P, ctypes.c_float, S, P]
    hw.hw_sum_f32.argtypes = [P, S, P, P]
    hw.hw_exscan_f32.argtypes = [P, P, S, P]
    n = 1 << args.log2n
    x, y, o, r = (ctx.vector(n=n, dtype=np.float32) for _ in range(4))
    x.fill(np.float32(0.5))
    y.fill(np.float32(0.25))
    px, py, po = x.device_ptr()[0], y.device_ptr()[0], o.device_ptr()[0]
    tmp = torch.empty(1, dtype=torch.float32, device="cuda")
    sp = ctx.stream(0)
    a = np.float32(2.5)
    pairs = {
        "map": (lambda: ctx.map(MAP_F32, x, o), lambda: hw.hw_map_f32(px, po, n, sp)),
        "zip": (lambda: ctx.zip(SAXPY_F32, x, y, o, args=[a]), lambda: hw.hw_saxpy_f32(px, py, po, 2.5, n, sp)),
        "reduce": (lambda: ctx.reduce_to(SUM_F32, x, r), lambda: hw.hw_sum_f32(px, n, tmp.data_ptr(), sp)),
        "scan": (lambda: ctx.scan(SUM_F32, x, o, np.float32(0)), lambda: hw.hw_exscan_f32(px, po, n, sp)),
    }
    res = {}
    for name, (fs, fh) in pairs.items():
        times = []
        for fn in (fs, fh):
            for _ in range(3):
                fn()
            ctx.sync()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(stream)
            for _ in range(10):
                fn()
            e1.record(stream)
            ctx.sync()
            times.append(e0.elapsed_time(e1) / 10)
        res[name] = {"skeleton_ms": round(times[0], 4), "handwritten_ms": round(times[1], 4),
                     "skeleton_over_handwritten": round(times[0] / times[1], 4)}
    res["handwritten"] = "nvcc float4 grid-stride kernels (map, saxpy), block-reduce + atomicAdd (sum, any order), " \
                         "CUB DeviceScan::ExclusiveSum (scan)"
    for v in (x, y, o, r):
        v.destroy()
    # disk cache: build from source vs load (fresh cache directory)
    srcs = [("map", MAP_F32), ("zip", SAXPY_F32), ("reduce", SUM_F32)]
    with tempfile.TemporaryDirectory() as d:
        c1 = skel.Context(1)
        c1.set_cache_dir(d)
        for k, src in srcs:
            c1.prepare(k, src)
        st1 = c1.stats()
        c1.close()
        c2 = skel.Context(1)
        c2.set_cache_dir(d)
        for k, src in srcs:
            c2.prepare(k, src)
        st2 = c2.stats()
        c2.close()
    res["kernel_cache"] = {"nvrtc_build_ms": round(st1["compile_ms"], 1), "disk_load_ms": round(st2["disk_load_ms"], 2),
                           "load_speedup": round(st1["compile_ms"] / max(st2["disk_load_ms"], 1e-6), 1),
                           "kernels": [k for k, _ in srcs], "paper": "loading is at least 5x faster (P:L248-250)"}
    res["small"] = bench_overhead_small(ctx, hw, stream)
    return res


def bench_overhead_small(ctx, hw, stream):
    """Latency-sized vectors: us per launch of each skeleton
    and of the same operation hand-written / from CUB, every launch replayed in
    a CUDA graph over rotating operand sets (>= 4x L2 of operands, so every
    launch reads from HBM), float32."""
    import math

    import torch
    from paper_conf_ipps_steuwerkg11_b200.workloads import MAP_F32, SAXPY_F32, SUM_F32
    import ctypes
    hw.hw_cubsum_f32.argtypes = [ctypes.c_void_p, ctypes.c_size_t, ctypes.c_void_p, ctypes.c_void_p]
    sp = ctx.stream(0)
    out = {}
    for k in (20, 22, 24):
        n = 1 << k
        R = max(2, min(64, math.ceil(4 * 126e6 / (2 * n * 4))))
        sets = []
        for _ in range(R):
            x, o, r = (ctx.vector(n=n if i < 2 else 1, dtype=np.float32) for i in range(3))
            x.fill(np.float32(1))
            sets.append((x, o, r, x.device_ptr()[0], o.device_ptr()[0], r.device_ptr()[0]))
        ops = {
            "map": (lambda st: ctx.map(MAP_F32, st[0], st[1]), lambda st: hw.hw_map_f32(st[3], st[4], n, sp)),
            "zip": (lambda st: ctx.zip(SAXPY_F32, st[0], st[1], st[1], args=[np.float32(2.5)]),
                    lambda st: hw.hw_saxpy_f32(st[3], st[4], st[4], 2.5, n, sp)),
            "reduce": (lambda st: ctx.reduce_to(SUM_F32, st[0], st[2]), lambda st: hw.hw_cubsum_f32(st[3], n, st[5], sp)),
            "scan": (lambda st: ctx.scan(SUM_F32, st[0], st[1], np.float32(0)),
                     lambda st: hw.hw_exscan_f32(st[3], st[4], n, sp)),
        }
        row = {}
        for name, pair in ops.items():
            us = []
            for op in pair:
                def fn(op=op):
                    for st in sets:
                        op(st)
                for _ in range(TUNE):
                    fn()
                ctx.sync()
                g = ctx.capture(fn)
                g.launch()
                ctx.sync()
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                e0.record(stream)
                for _ in range(10):
                    g.launch()
                e1.record(stream)
                ctx.sync()
                g.destroy()
                us.append(round(e0.elapsed_time(e1) * 1e3 / (10 * R), 2))
            row[name] = {"skeleton_us": us[0], "reference_us": us[1]}
        out[f"2^{k}"] = row
        for st in sets:
            for v in st[:3]:
                v.destroy()
    out["reference"] = "map/zip: hand-written float4 nvcc kernels; reduce: CUB DeviceReduce::Sum (two kernels, " \
                       "commutative only); scan: CUB DeviceScan::ExclusiveSum"
    return out


FP32_NOMINAL_OPS = 148 * 128 * 1.965e9  # nominal: 148 SMs x 128 FP32 lanes x 1.965 GHz
MANDEL_BLOCK = 128  # CTA size of the Mandelbrot Maps (skel_set_block_size; measured best)


def bench_mandelbrot(ctx, skel, stream, world, rank, barrier, max_over_ranks, args):
    """configs[2]: 4096x3072, cap 256, rows block-distributed over the GPUs --
    the paper's Map over positions and the NEXT-4 variants (all bit-identical
    to eq. (5) as written, tests/test_gpu_mandelbrot.py): index Map, blocked
    loop control, pixel pairs with packed FP32x2, exact periodicity checking,
    cyclic rows; the cap-4096 heavy variant; configs[0] 1024x768 on one GPU.
    FP32 fraction = 8 FP32 operations per iteration AS WRITTEN x sum of the
    counts / time / FP32 lane peak MEASURED in this run by a probe Map
    (workloads/probe_fp32.cu: independent packed FP32 adds on every lane; the
    nominal 148 x 128 x 1.965 GHz is reported beside it).  The periodicity
    variants execute fewer iterations than that sum: their figure is an
    algorithmic-equivalent rate, not pipe utilisation."""
    W, H, cap = 4096, 3072, 256
    reps = max(args.steps, 10)
    ctx.set_block_size(MANDEL_BLOCK)
    try:
        return _bench_mandelbrot(ctx, skel, stream, world, rank, barrier, max_over_ranks, reps, W, H, cap)
    finally:
        ctx.set_block_size(0)


def _bench_mandelbrot(ctx, skel, stream, world, rank, barrier, max_over_ranks, reps, W, H, cap):
    import torch
    import skel_inputs as si
    from paper_conf_ipps_steuwerkg11_b200.mandelbrot import CyclicMandelbrot
    from paper_conf_ipps_steuwerkg11_b200.workloads import (MANDELBROT, MANDELBROT_BLOCKED, MANDELBROT_INDEX,
                                                            MANDELBROT_PAIRS, MANDELBROT_PERIODIC, PROBE_FP32,
                                                            PROBE_FP32_OPS_PER_STEP)

    def timed(fn, n=reps):
        """GPU time per call: the call captured once as a CUDA graph and replayed
        n times (a 25 us launch timed eagerly would measure the Python/ctypes call
        rate); eager calls where graphs are unavailable."""
        for _ in range(3):
            fn()
        ctx.sync()
        run, g = fn, None
        if not os.environ.get("SKEL_BENCH_NO_GRAPH"):
            try:
                g = ctx.capture(fn)
                g.launch()
                ctx.sync()
                run = g.launch
            except skel.SkelError:
                g, run = None, fn
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        barrier()
        torch.cuda.synchronize()
        e0.record(stream)
        for _ in range(n):
            run()
        e1.record(stream)
        ctx.sync()
        if g is not None:
            g.destroy()
        return max_over_ranks(e0.elapsed_time(e1) / n)

    # the FP32 lane peak, measured: every GPU runs the probe Map over 4 resident
    # waves of threads (16 FP32 operations per step and thread)
    sms = torch.cuda.get_device_properties(torch.cuda.current_device()).multi_processor_count
    npr, steps = sms * 2048 * 4 * world, 2048
    pv = ctx.vector(n=npr, dtype=np.float32)
    if world > 1:
        pv.set_distribution(skel.BLOCK)
    ms_p = timed(lambda: ctx.map_index(PROBE_FP32, npr, pv, args=[np.float32(1e-7), np.int32(steps)]), n=5)
    pv.destroy()
    peak = (npr // world) * steps * PROBE_FP32_OPS_PER_STEP / (ms_p * 1e-3)  # per GPU
    peak_all = peak * world
    pos = si.mandelbrot_positions(W, H)
    vin = ctx.vector(n=pos.size, dtype=pos.dtype)
    pairs = pos.view(si.POS2_DTYPE)
    vin2 = ctx.vector(n=pairs.size, dtype=pairs.dtype)
    if world > 1:
        vin.set_distribution(skel.BLOCK)
        vin2.set_distribution(skel.BLOCK)
    lo, hi = vin.part(rank) if world > 1 else (0, pos.size)
    vin.upload_part(lo, pos[lo:hi])
    lo2, hi2 = vin2.part(rank) if world > 1 else (0, pairs.size)
    vin2.upload_part(lo2, pairs[lo2:hi2])
    out = ctx.vector(n=pos.size, dtype=np.int32)
    out2 = ctx.vector(n=pairs.size, dtype=si.CNT2_DTYPE)
    oi = ctx.vector(n=pos.size, dtype=np.int32)
    if world > 1:
        oi.set_distribution(skel.BLOCK)
    capv = np.int32(cap)
    ms = {}
    ms["paper"] = timed(lambda: ctx.map(MANDELBROT, vin, out, args=[capv]))
    counts = out.download()  # collective in rank mode: every rank takes part
    ms["index_map"] = timed(lambda: ctx.map_index(MANDELBROT_INDEX, W * H, oi, args=[np.int32(W), np.int32(H), capv]))
    ms["blocked"] = timed(lambda: ctx.map(MANDELBROT_BLOCKED, vin, out, args=[capv]))
    same = np.array_equal(out.download(), counts)
    ms["pairs"] = timed(lambda: ctx.map(MANDELBROT_PAIRS, vin2, out2, args=[capv]))
    same &= np.array_equal(out2.download().view(np.int32), counts)
    ms["periodic"] = timed(lambda: ctx.map(MANDELBROT_PERIODIC, vin, out, args=[capv]))
    same &= np.array_equal(out.download(), counts)
    from paper_conf_ipps_steuwerkg11_b200.workloads import MANDELBROT_PAIRS_PERIODIC
    ms["pairs_periodic"] = timed(lambda: ctx.map(MANDELBROT_PAIRS_PERIODIC, vin2, out2, args=[capv]))
    same &= np.array_equal(out2.download().view(np.int32), counts)
    # cyclic rows (device k: rows k, k+D, ...): the compute step alone and the
    # whole image on device 0 (gather + un-permute)
    cm = CyclicMandelbrot(ctx, W, H)
    ms["cyclic_compute"] = timed(lambda: cm.compute(cap))
    ms["cyclic_image"] = timed(lambda: cm.image(cap))
    same &= np.array_equal(cm.counts(cap), counts)
    iters = int(counts.astype(np.int64).sum())
    res = {"config": "configs[2]: 4096x3072, cap 256, block rows", "ms": ms["paper"],
           "Mpix_per_s": W * H / (ms["paper"] * 1e-3) / 1e6, "variants_ms": ms,
           "all_bit_identical": bool(same), "sum_iter": iters,
           "Giter_per_s": iters / (ms["paper"] * 1e-3) / 1e9,
           "fp32_peak": {"value": peak_all, "per_gpu": peak, "unit": "FP32 ops/s",
                         "source": "measured in this run: probe Map workloads/probe_fp32.cu (8 independent chains of "
                                   "add.rn.f32x2 per thread, 4 resident waves)",
                         "nominal_per_gpu": FP32_NOMINAL_OPS, "measured_over_nominal": peak / FP32_NOMINAL_OPS},
           "cta_threads": MANDEL_BLOCK,
           "fp32_frac": {k: 8 * iters / (v * 1e-3) / peak_all for k, v in ms.items()
                         if not k.startswith("cyclic_image")}}
    # heavy variant ("also report the cap-4096 variant")
    c4 = np.int32(4096)
    heavy = {}
    for name, fn, vi, vo in (("paper", MANDELBROT, vin, out), ("blocked", MANDELBROT_BLOCKED, vin, out),
                             ("periodic", MANDELBROT_PERIODIC, vin, out)):
        heavy[name] = timed(lambda: ctx.map(fn, vi, vo, args=[c4]), n=3)
    it4096 = int(out.download().astype(np.int64).sum())
    # 8x4 tiles per warp with periodicity checking: a void index Map writing the image
    from paper_conf_ipps_steuwerkg11_b200.workloads import MANDELBROT_TILES_PERIODIC
    img = ctx.vector(n=pos.size, dtype=np.int32)
    img.fill_dist(skel.COPY if world > 1 else skel.SINGLE, np.int32(0))
    heavy["tiles_periodic"] = timed(lambda: ctx.map_index(MANDELBROT_TILES_PERIODIC, W * H, None,
                                                          args=[img, np.int32(W), np.int32(H), c4]), n=3)
    img.destroy()
    res["cap4096"] = {"sum_iter": it4096, "ms": heavy,
                      "fp32_frac": {k: 8 * it4096 / (v * 1e-3) / peak_all for k, v in heavy.items()},
                      "note": "periodic variants stop a member once its orbit repeats bit for bit: their fraction "
                              "is algorithmic-equivalent (sum of the counts x 8 / time), not pipe utilisation"}
    for v in (vin, vin2, out, out2, oi):
        v.destroy()
    # configs[0]: 1024x768, cap 256, single distribution (device 0 / rank 0)
    ps = si.mandelbrot_positions(1024, 768)
    vs = ctx.vector(n=ps.size, dtype=ps.dtype)
    vs.set_distribution(skel.SINGLE)
    vs.upload(ps)
    os_ = ctx.vector(n=ps.size, dtype=np.int32)
    os_.set_distribution(skel.SINGLE)
    ps2 = ps.view(si.POS2_DTYPE)
    vs2 = ctx.vector(n=ps2.size, dtype=ps2.dtype)
    vs2.set_distribution(skel.SINGLE)
    vs2.upload(ps2)
    os2 = ctx.vector(n=ps2.size, dtype=si.CNT2_DTYPE)
    os2.set_distribution(skel.SINGLE)
    ms0 = {"paper": timed(lambda: ctx.map(MANDELBROT, vs, os_, args=[capv])),
           "pairs": timed(lambda: ctx.map(MANDELBROT_PAIRS, vs2, os2, args=[capv])),
           "periodic": timed(lambda: ctx.map(MANDELBROT_PERIODIC, vs, os_, args=[capv]))}
    res["configs0_1024x768"] = {"ms": ms0["paper"], "variants_ms": ms0,
                                "Mpix_per_s": ps.size / (ms0["paper"] * 1e-3) / 1e6, "sum_iter": 28347768,
                                "fp32_frac": {k: 8 * 28347768 / (v * 1e-3) / peak for k, v in ms0.items()},
                                "note": "single distribution: one GPU computes, 2.6 waves (latency-sized)"}
    for v in (vs, os_, vs2, os2):
        v.destroy()
    return res


_LM_CACHE: dict = {}


def lm_subsets(nev, nsub, lo, hi):
    """Events [lo, hi) of subsets 0..nsub-1 of nev events each (generated once per job)."""
    import skel_inputs as si
    out = []
    for l in range(nsub):
        if (nev, l) not in _LM_CACHE:
            _LM_CACHE[(nev, l)] = si.lmosem_events(nev, subset=l)
        out.append(_LM_CACHE[(nev, l)][lo:hi])
    return out


def bench_lmosem(ctx, skel, stream, world, rank, barrier, max_over_ranks, args):
    """configs[3]/[4]: one subset of 10^6 events into 150x150x280, events
    block-distributed; the error-image Map in the form lmosem.LMOSEM.plan picks
    for 10^6/N events per GPU (a lanes Map with 4 threads per event in the
    given order).  `device_order`: the same subset with every GPU's events
    reordered by path length ON THE DEVICE first (counting Map + Scan +
    scattering Map, included in the time)."""
    import torch
    from paper_conf_ipps_steuwerkg11_b200.lmosem import LMOSEM
    nev = 1_000_000
    ev = lm_subsets(nev, 1, 0, nev)[0]
    rec = LMOSEM(ctx)
    rec.prepare()
    evv = ctx.vector(n=nev, dtype=ev.dtype)
    if world > 1:
        evv.set_distribution(skel.BLOCK)
    lo, hi = evv.part(rank) if world > 1 else (0, nev)
    evv.upload_part(lo, ev[lo:hi])
    for _ in range(TUNE):
        rec.subset(evv)
    ctx.sync()
    reps = 10

    def timed(fn):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        barrier()
        torch.cuda.synchronize()
        e0.record(stream)
        for _ in range(reps):
            fn()
        e1.record(stream)
        ctx.sync()
        return max_over_ranks(e0.elapsed_time(e1) / reps)

    ms = timed(lambda: rec.subset(evv))
    for _ in range(TUNE):
        rec.subset(evv, fused=True)
    ms_fused = timed(lambda: rec.subset(evv, fused=True))
    # the two fixed orders the default (order="auto") chooses between
    recg = LMOSEM(ctx, order="given")
    recg.prepare()
    for _ in range(TUNE):
        recg.subset(evv)
    ms_given = timed(lambda: recg.subset(evv))
    try:
        if os.environ.get("SKEL_BENCH_NO_GRAPH"):
            raise skel.SkelError(8, "graphs disabled")
        g = ctx.capture(lambda: rec.subset(evv))  # the subset loop body as one CUDA graph
        ms_graph = timed(g.launch)
        g.destroy()
    except skel.SkelError:  # a collective backend that cannot be captured
        ms_graph = ms
    # the same subset with the events ordered on the device (sort inside the time)
    recd = LMOSEM(ctx, order="device")
    recd.prepare()
    for _ in range(TUNE):
        recd.subset(evv)
    ms_dev = timed(lambda: recd.subset(evv))
    ms_sort = timed(lambda: recd.order_on_device(evv))
    try:  # the same as CUDA graphs: GPU time without the per-call host overhead
        if os.environ.get("SKEL_BENCH_NO_GRAPH"):
            raise skel.SkelError(8, "graphs disabled")
        g = ctx.capture(lambda: recd.subset(evv))
        ms_dev_graph = timed(g.launch)
        g.destroy()
        g = ctx.capture(lambda: recd.order_on_device(evv))
        ms_sort_graph = timed(g.launch)
        g.destroy()
    except skel.SkelError:
        ms_dev_graph, ms_sort_graph = ms_dev, ms_sort
    coll = None
    if world > 1:  # the exchange steps alone, bus GB/s vs NVLink
        S = rec.nvox * 4
        c, f = rec.c, rec.f

        def fill_rs():
            c.fill_dist(skel.COPY, np.float32(0))
            c.set_distribution(skel.BLOCK, skel.COMBINE_ADD)  # copy -> block + add: reduce-scatter

        def ag():
            f.set_distribution(skel.BLOCK)  # copy -> block: local slice (no data movement)
            f.set_distribution(skel.COPY)   # block -> copy: all-gather
        ms_fill = timed(lambda: c.fill_dist(skel.COPY, np.float32(0)))
        ms_rs = max(timed(fill_rs) - ms_fill, 1e-6)
        ms_ag = timed(ag)
        busf = (world - 1) / world
        coll = {"bytes": S, "reduce_scatter_ms": ms_rs, "all_gather_ms": ms_ag,
                "reduce_scatter_busbw_GBps": S * busf / (ms_rs * 1e-3) / 1e9,
                "all_gather_busbw_GBps": S * busf / (ms_ag * 1e-3) / 1e9,
                "peak_GBps": 770.0, "peak_source": "B200_PROFILING.md measured peer copy per direction "
                                                  "(900 nominal)"}
    roof = lmosem_roofline(ctx, skel, recg, recd, evv, timed, world)
    evv.destroy()
    # configs[4]: the full reconstruction -- 10 subsets of 10^6 events (10^7,
    # P:L603-605), each subset a different synthetic draw, all events staged on
    # the devices beforehand (240 MB); one pass over the subsets from f0 = 1
    nsub = 10
    full = {}
    subs = []
    for evl in lm_subsets(nev, nsub, lo, hi):
        v = ctx.vector(n=nev, dtype=evl.dtype)
        if world > 1:
            v.set_distribution(skel.BLOCK)
        v.upload_part(lo, evl)
        subs.append(v)
    for mode in ("auto", "given"):
        rec2 = LMOSEM(ctx, order=mode)
        rec2.prepare()
        for v in subs:  # stage every subset (lazy H2D) and warm up
            rec2.subset(v)
        ctx.sync()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        barrier()
        torch.cuda.synchronize()
        e0.record(stream)
        rec2.f.fill_dist(skel.BLOCK, np.float32(1))
        for v in subs:
            rec2.subset(v)
        e1.record(stream)
        ctx.sync()
        full[mode] = max_over_ranks(e0.elapsed_time(e1))
    for v in subs:
        v.destroy()
    per = -(-nev // world)
    src, lanes = rec.plan(per)
    return {"config": "configs[3]/[4]: one subset, 10^6 events, 150x150x280, events block over GPUs",
            "subset_s": ms * 1e-3, "subset_s_graph": ms_graph * 1e-3, "subset_s_fused": ms_fused * 1e-3,
            "policy": {"order": "device" if rec.ordered(per) else "given", "lanes": lanes, "cta_threads": 128,
                       "events_per_gpu": per},
            "roofline": roof, "exchange": coll,
            "events_per_s": nev / (min(ms, ms_graph, ms_fused) * 1e-3),
            "full_recon_s": full["auto"] * 1e-3, "full_recon": "10 subsets x 10^6 events (configs[4]), f0 = 1, "
                                                               "events resident on the devices",
            "given_order": {"subset_s": ms_given * 1e-3, "full_recon_s": full["given"] * 1e-3,
                            "map_lanes": recg.plan(per)[1]},
            "device_order": {"subset_s": ms_dev * 1e-3, "order_s": ms_sort * 1e-3,
                             "subset_s_graph": ms_dev_graph * 1e-3, "order_s_graph": ms_sort_graph * 1e-3,
                             "map_lanes": recd.plan(-(-nev // world))[1],
                             "note": "every GPU's events reordered by path length on the device (lmosem_order.cu: "
                                     "counting Map + Scan + scattering Map, inside the timed subset) before the "
                                     "error-image Map; same image up to float rounding (R10(x))"},
            "note": "includes f all-gather, c zero-fill, Siddon Map, c reduce-scatter and update Zip; "
                    "subset_s = eager calls, subset_s_graph = the same subset replayed as a CUDA graph, "
                    "subset_s_fused = the tail as one peer-memory kernel (skel_zip_combine, NEXT-1)"}


def lmosem_l1_hit():
    """L1 hit rate of the forward-projection gathers of the error-image Map,
    from the committed ncu capture (profiles/lmosem_l1.json), or None."""
    try:
        with open(os.path.join(ROOT, "profiles", "lmosem_l1.json")) as fh:
            return json.load(fh)
    except Exception:
        return None


def lmosem_roofline(ctx, skel, rec, recd, evv, timed, nd):
    """Roofline of the error-image Map.  Every voxel visit of a
    path is one scattered 4-byte request in each walk (a gather of f forward,
    a red.add into c backward) and the lanes of a warp are on different rays,
    so the Map is bound by how fast the SMs' L1TEX units can issue scattered
    requests to L2.  The peaks are measured in the same run by probe Maps
    (workloads/probe_*.cu) issuing random scattered gathers / vector
    reductions; a gather costs h/peak_resident + (1-h)/peak_image with h the
    Map's measured L1 hit rate (profiles/lmosem_l1.json, ncu); the Map's ideal
    time is V x that + R/peak_red_v4 for V voxel visits and R vector
    reductions (4-float groups entered), both counted by Maps over the same
    events."""
    from paper_conf_ipps_steuwerkg11_b200.workloads import (LMOSEM_GROUPS, LMOSEM_VISITS, PROBE_GATHER, PROBE_K,
                                                            PROBE_SCATTER_RED, PROBE_SCATTER_RED4, SUM_I32)
    dims = rec.dims_args
    nvis = ctx.vector(n=evv.n, dtype=np.int32)
    if evv.distribution == skel.BLOCK:
        nvis.set_distribution(skel.BLOCK)
    ctx.map(LMOSEM_VISITS, evv, nvis, args=dims)
    visits = int(ctx.reduce(SUM_I32, nvis))  # all ranks' events
    ctx.map(LMOSEM_GROUPS, evv, nvis, args=dims)
    groups = int(ctx.reduce(SUM_I32, nvis))  # vector reductions of the back projection
    nvis.destroy()
    f, c = rec.f, rec.c
    f.set_distribution(skel.COPY)
    c.fill_dist(skel.COPY, np.float32(0))
    for _ in range(TUNE):
        rec.error_map(evv)
    ms_map = timed(lambda: rec.error_map(evv))
    recd.f.set_distribution(skel.COPY)
    recd.c.fill_dist(skel.COPY, np.float32(0))
    evo = recd.order_on_device(evv)
    for _ in range(TUNE):
        recd.error_map(evo)
    ms_map_ord = timed(lambda: recd.error_map(evo))
    c.mark_device_modified()
    recd.c.mark_device_modified()
    # probes: 2^20 elements x PROBE_K scattered requests each (per GPU), into (a) an
    # image-sized 25 MB buffer (random lines: L2 hit/miss and far-partition traffic
    # included) and (b) a small buffer (64 KB gathers: L1-resident; 1 MB reductions:
    # L2-resident), which isolates the SM's rate of issuing scattered requests
    npr = 1 << 20
    idx = ctx.vector(np.arange(npr, dtype=np.uint32))
    img = ctx.vector(n=rec.nvox, dtype=np.float32)  # whole buffers on every GPU (copy)
    img.fill_dist(skel.COPY, np.float32(1))
    acc = ctx.vector(n=rec.nvox, dtype=np.float32)
    acc.fill_dist(skel.COPY, np.float32(0))
    gout = ctx.vector(n=npr, dtype=np.float32)
    probes = {}
    for tag, ng, nr in (("image", rec.nvox, rec.nvox), ("resident", 1 << 14, 1 << 18)):
        ng, nr = np.uint32(ng), np.uint32(nr)
        for _ in range(TUNE):
            ctx.map(PROBE_GATHER, idx, gout, args=[img, ng])
            ctx.map(PROBE_SCATTER_RED, idx, None, args=[acc, nr])
            ctx.map(PROBE_SCATTER_RED4, idx, None, args=[acc, nr])
        ms_g = timed(lambda: ctx.map(PROBE_GATHER, idx, gout, args=[img, ng]))
        ms_r = timed(lambda: ctx.map(PROBE_SCATTER_RED, idx, None, args=[acc, nr]))
        ms_r4 = timed(lambda: ctx.map(PROBE_SCATTER_RED4, idx, None, args=[acc, nr]))
        probes[tag] = tuple(npr * PROBE_K / (t * 1e-3) / 1e9 for t in (ms_g, ms_r, ms_r4))
    for v in (idx, img, acc, gout):
        v.destroy()
    peak_r4 = max(p[2] for p in probes.values())
    l1 = lmosem_l1_hit()
    h = float(l1["given"]["l1_hit_rate"]) if l1 else None
    hd = float(l1["device"]["l1_hit_rate"]) if l1 and "device" in l1 else h
    g_res, g_img = probes["resident"][0], probes["image"][0]

    def gather_rate(hit):  # G gathers/s at L1 hit rate `hit` (None: the resident probe, an upper bound)
        if hit is None:
            return g_res
        return 1.0 / (hit / g_res + (1.0 - hit) / g_img)
    pg, pgd = gather_rate(h), gather_rate(hd)
    # requests of the Map: one gather per visit (forward), one vector reduction per
    # 4-float group entered (back projection); ideal = each at its measured peak
    reqs = (visits + groups) / nd
    ideal_ms = (visits / nd) / (pg * 1e9) * 1e3 + (groups / nd) / (peak_r4 * 1e9) * 1e3
    # device order: the forward projection gathers 16 bytes per 4-float group
    ideal_ord_ms = (groups / nd) / (pgd * 1e9) * 1e3 + (groups / nd) / (peak_r4 * 1e9) * 1e3
    return {"kernel": "LM OSEM error-image Map (skel_ew_kernel, lanes Map + lmosem_lanes)", "bound": "l1tex",
            "achieved": reqs / (ms_map * 1e-3) / 1e9, "peak": reqs / (ideal_ms * 1e-3) / 1e9,
            "unit": "G scattered requests/s per GPU",
            "frac": ideal_ms / ms_map, "map_ms": ms_map, "ideal_ms": ideal_ms, "visits_per_subset": visits,
            "l1_hit_rate": h, "gather_rate_G_per_s": pg,
            "device_order": {"map_ms": ms_map_ord, "frac": ideal_ord_ms / ms_map_ord, "ideal_ms": ideal_ord_ms,
                             "l1_hit_rate": hd,
                             "note": "the Map over the device-ordered events with the prepared function (one 16-byte "
                                     "gather per 4-float group forward, one red.v4 per group backward): 2 x groups "
                                     "requests"},
            "vector_reductions_per_subset": groups, "peak_red_v4": peak_r4, "peak_red": max(p[1] for p in probes.values()),
            "probes_Greq_per_s": {k: {"gather": v[0], "red": v[1], "red_v4": v[2]} for k, v in probes.items()},
            "peak_source": "measured in this run: probe Maps workloads/probe_gather.cu, probe_scatter.cu, "
                           "probe_scatter4.cu (random 4-byte gathers / red.add.f32 / red.add.v4.f32, 32 lanes on "
                           "32 lines) into a 25 MB image-sized buffer and an L1/L2-resident one; the gather rate "
                           "is the two probes' rates weighted by the Map's ncu L1 hit rate (profiles/lmosem_l1.json; "
                           "absent: the resident probe, an upper bound)"}


if __name__ == "__main__":
    main()
