"""Time the Mandelbrot Maps (paper form, blocked form) at 4096x3072, cap 256 and 4096."""
import json, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import MANDELBROT, MANDELBROT_BLOCKED, MANDELBROT_PAIRS

pos = si.mandelbrot_positions(4096, 3072)
with skel.Context(1) as ctx:
    st = torch.cuda.ExternalStream(ctx.stream(0))
    vin = ctx.vector(pos)
    vin2 = ctx.vector(pos.view(si.POS2_DTYPE))
    res = {"defines": os.environ.get("SKEL_NVRTC_DEFINES", "")}
    for cap in (256, 4096):
        outs = {}
        for name, fn in (("paper", MANDELBROT), ("blocked", MANDELBROT_BLOCKED), ("pairs", MANDELBROT_PAIRS)):
            v = vin2 if name == "pairs" else vin
            out = ctx.vector(n=v.n, dtype=si.CNT2_DTYPE if name == "pairs" else np.int32)
            for _ in range(2):  # first launch decides the grid policy on a sample
                ctx.map(fn, v, out, args=[np.int32(cap)])
            ctx.sync()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(st)
            for _ in range(10):
                ctx.map(fn, v, out, args=[np.int32(cap)])
            e1.record(st)
            ctx.sync()
            res[f"{name}_{cap}_ms"] = round(e0.elapsed_time(e1) / 10, 4)
            outs[name] = out.download().view(np.int32)
        res[f"same_{cap}"] = bool(np.array_equal(outs["paper"], outs["blocked"])) and \
            bool(np.array_equal(outs["paper"], outs["pairs"]))
        res[f"iters_{cap}"] = int(outs["paper"].astype(np.int64).sum())
    print(json.dumps(res))
