"""Run the Mandelbrot Map and one LM OSEM subset (for ncu captures)."""
import sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.lmosem import LMOSEM
from paper_conf_ipps_steuwerkg11_b200.workloads import MANDELBROT

which = sys.argv[1] if len(sys.argv) > 1 else "both"
with skel.Context(1) as ctx:
    if which in ("both", "mandel"):
        pos = si.mandelbrot_positions(4096, 3072)
        vin = ctx.vector(pos)
        out = ctx.vector(n=pos.size, dtype=np.int32)
        for _ in range(3):
            ctx.map(MANDELBROT, vin, out, args=[np.int32(256)])
        ctx.sync()
    if which in ("both", "lmosem", "lmosem_device"):
        ev = si.lmosem_events(1_000_000, subset=0)
        rec = LMOSEM(ctx, order="device" if which == "lmosem_device" else "given")
        evv = rec.events(ev)
        for _ in range(3):
            rec.subset(evv)
        ctx.sync()
print("done")
