"""Small-size Reduce / Scan / Map: skeleton kernels vs CUB and hand-written
nvcc kernels on the same buffers, each replayed as a CUDA graph of R
back-to-back launches over rotating operand sets (R x footprint >= 4x L2, as
in bench.py's sweep).  Prints one JSON line per size (us per launch).

usage: python tools/small_n_probe.py [log2n ...]
"""
import ctypes
import json
import math
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import numpy as np  # noqa: E402
import torch  # noqa: E402

from paper_conf_ipps_steuwerkg11_b200 import skel  # noqa: E402
from paper_conf_ipps_steuwerkg11_b200.workloads import MAP_F32, SAXPY_F32, SUM_F32  # noqa: E402


def main():
    ks = [int(a) for a in sys.argv[1:]] or [18, 20, 21, 22, 23, 24, 26]
    hw = ctypes.CDLL(os.path.join(ROOT, "paper_conf_ipps_steuwerkg11_b200", "libhandwritten.so"))
    P, S = ctypes.c_void_p, ctypes.c_size_t
    hw.hw_map_f32.argtypes = [P, P, S, P]
    hw.hw_saxpy_f32.argtypes = [P, P, P, ctypes.c_float, S, P]
    hw.hw_sum_f32.argtypes = [P, S, P, P]
    hw.hw_cubsum_f32.argtypes = [P, S, P, P]
    hw.hw_exscan_f32.argtypes = [P, P, S, P]
    l2 = 126e6
    with skel.Context(1) as ctx:
        sp = ctx.stream(0)
        stream = torch.cuda.ExternalStream(sp)
        for k in ks:
            n = 1 << k
            R = max(2, min(128, math.ceil(4 * l2 / (2 * n * 4))))
            sets = []
            for _ in range(R):
                x, o, r = ctx.vector(n=n, dtype=np.float32), ctx.vector(n=n, dtype=np.float32), \
                    ctx.vector(n=1, dtype=np.float32)
                x.fill(np.float32(1))
                o.fill(np.float32(0))
                r.fill(np.float32(0))
                sets.append((x, o, r, x.device_ptr()[0], o.device_ptr()[0], r.device_ptr()[0]))
            ops = {
                "map_skel": lambda st: ctx.map(MAP_F32, st[0], st[1]),
                "zip_skel": lambda st: ctx.zip(SAXPY_F32, st[0], st[1], st[1], args=[np.float32(2.5)]),
                "zip_hw": lambda st: hw.hw_saxpy_f32(st[3], st[4], st[4], 2.5, n, sp),
                "map_hw": lambda st: hw.hw_map_f32(st[3], st[4], n, sp),
                "reduce_skel": lambda st: ctx.reduce_to(SUM_F32, st[0], st[2]),
                "reduce_cub": lambda st: hw.hw_cubsum_f32(st[3], n, st[5], sp),
                "reduce_atomic": lambda st: hw.hw_sum_f32(st[3], n, st[5], sp),
                "scan_skel": lambda st: ctx.scan(SUM_F32, st[0], st[1], np.float32(0)),
                "scan_cub": lambda st: hw.hw_exscan_f32(st[3], st[4], n, sp),
            }
            if os.environ.get("PROBE_OPS"):
                keep = os.environ["PROBE_OPS"].split(",")
                ops = {k2: v for k2, v in ops.items() if any(k2.startswith(p) for p in keep)}
            row = {"log2n": k, "R": R}
            for name, op in ops.items():
                def fn(op=op):
                    for st in sets:
                        op(st)
                fn()
                ctx.sync()
                g = ctx.capture(fn)
                g.launch()
                ctx.sync()
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                reps = 20
                e0.record(stream)
                for _ in range(reps):
                    g.launch()
                e1.record(stream)
                ctx.sync()
                g.destroy()
                row[name] = round(e0.elapsed_time(e1) * 1e3 / (reps * R), 2)
            # correctness spot check of the skeleton results
            ctx.reduce_to(SUM_F32, sets[0][0], sets[0][2])
            row["reduce_ok"] = float(sets[0][2].download()[0]) == float(n)
            ctx.scan(SUM_F32, sets[0][0], sets[0][1], np.float32(0))
            y = sets[0][1].download()
            row["scan_ok"] = bool(y[0] == 0 and y[-1] == n - 1 and y[n // 3] == n // 3) if n <= 1 << 24 else None
            print(json.dumps(row), flush=True)
            for st in sets:
                for v in st[:3]:
                    v.destroy()


if __name__ == "__main__":
    main()
