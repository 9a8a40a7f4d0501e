"""Per-GPU work of LM OSEM at D GPUs, measured on one GPU: the error-image
Map over 10^6/D events (what each GPU runs per subset at D GPUs), plus the
other per-subset kernels.  Prints ms per Map for D = 1, 2, 4, 8."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch

import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import LMOSEM_ERROR

if os.environ.get("LM_SRC"):  # A/B: an alternative error-image function text
    LMOSEM_ERROR = open(os.environ["LM_SRC"]).read()

ev = si.lmosem_events(1_000_000, subset=0)
with skel.Context(1) as ctx:
    stream = torch.cuda.ExternalStream(ctx.stream(0))
    f = ctx.vector(n=150 * 150 * 280, dtype=np.float32).fill(np.float32(1))
    c = ctx.vector(n=150 * 150 * 280, dtype=np.float32)
    dims = [np.int32(150), np.int32(150), np.int32(280)]
    for D in (1, 2, 4, 8):
        part = ev[: 1_000_000 // D]
        if os.environ.get("LM_ORDER") == "dealt":  # longest first, warp groups dealt to the CTAs
            from paper_conf_ipps_steuwerkg11_b200.lmosem import deal_warps
            part = deal_warps(part, block=int(os.environ.get("SKEL_BLOCK_SIZE", "256")))
        elif os.environ.get("LM_ORDER"):  # each GPU orders its part longest path first
            from paper_conf_ipps_steuwerkg11_b200.lmosem import order_by_path
            part = order_by_path(part)
        e = ctx.vector(part)
        for _ in range(3):
            ctx.map(LMOSEM_ERROR, e, None, args=[f, c, *dims])
        ctx.sync()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(stream)
        for _ in range(10):
            ctx.map(LMOSEM_ERROR, e, None, args=[f, c, *dims])
        e1.record(stream)
        ctx.sync()
        print(f"D={D} events={1_000_000 // D} map_ms={e0.elapsed_time(e1) / 10:.4f}", flush=True)
