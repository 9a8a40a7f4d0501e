"""One Mandelbrot Map variant on the paper image (4096x3072, cap 256), launched
a few times -- the target of an ncu capture (tools/run_*.sh).
usage: python tools/mandel_one.py <variant> [block]"""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200 import workloads as w

V = {"paper": w.MANDELBROT, "blocked": w.MANDELBROT_BLOCKED, "periodic": w.MANDELBROT_PERIODIC,
     "pairs": w.MANDELBROT_PAIRS, "pairs_periodic": w.MANDELBROT_PAIRS_PERIODIC}
name = sys.argv[1]
block = int(sys.argv[2]) if len(sys.argv) > 2 else 0
src = V[name]
pos = si.mandelbrot_positions(4096, 3072)
two = "pairs" in name
with skel.Context(1) as ctx:
    if block:
        ctx.set_block_size(block)
    vin = ctx.vector(pos.view(si.POS2_DTYPE) if two else pos)
    out = ctx.vector(n=vin.n, dtype=si.CNT2_DTYPE if two else np.int32)
    for _ in range(4):
        ctx.map(src, vin, out, args=[np.int32(256)])
    ctx.sync()
    print(name, int(out.download().view(np.int32).astype(np.int64).sum()))
