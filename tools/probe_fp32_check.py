import os, sys, time
sys.path.insert(0, os.getcwd())
import numpy as np, torch
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import PROBE_FP32
NV = PROBE_FP32.replace("asm volatile", "asm")
with skel.Context(1) as ctx:
    st = torch.cuda.ExternalStream(ctx.stream(0))
    for name, src in (("volatile", PROBE_FP32),):
        for block in (128, 256):
            for waves in (1, 4, 8):
                ctx.set_block_size(block)
                n = 148 * 2048 * waves
                v = ctx.vector(n=n, dtype=np.float32)
                steps = 2048
                f = lambda: ctx.map_index(src, n, v, args=[np.float32(1e-7), np.int32(steps)])
                for _ in range(3): f()
                ctx.sync()
                g = ctx.capture(f); g.launch(); ctx.sync()
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                e0.record(st)
                for _ in range(5): g.launch()
                e1.record(st); ctx.sync()
                ms = e0.elapsed_time(e1) / 5
                print(name, block, waves, f"{n*steps*16/(ms*1e-3)/1e12:.2f} T", flush=True)
                g.destroy(); v.destroy()
