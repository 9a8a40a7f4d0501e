"""A few Scans at 2^k float32 (default 22) -- an ncu target for the small-vector Scan path."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import SUM_F32
k = int(sys.argv[1]) if len(sys.argv) > 1 else 22
x = si.uniform_f32(1 << k, 1)
with skel.Context(1) as ctx:
    v = ctx.vector(x)
    o = ctx.vector(n=x.size, dtype=np.float32)
    for _ in range(6):
        ctx.scan(SUM_F32, v, o, np.float32(0))
    ctx.sync()
    print("ok", float(o.download()[-1]))
