"""Per-GPU error-image Map of LM OSEM at D GPUs, measured on one GPU: the Map
over 10^6/D events (one GPU's part of a subset at D GPUs) for the one-thread-
per-event Map and the lanes Map (skel_map_lanes, `lanes` threads per event,
workloads/lmosem_lanes.cu), in the given event order and longest-path-first
order, at CTA sizes 128/256.  One JSON line per point."""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch

import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.lmosem import LMOSEM
from paper_conf_ipps_steuwerkg11_b200.workloads import (LMOSEM_ERROR, LMOSEM_ERROR_PREPARED, LMOSEM_LANES,
                                                        LMOSEM_LANES_PREPARED)

if os.environ.get("LM_MINB"):  # register cap: minimum resident CTAs per SM for the lanes Map
    LMOSEM_LANES = f"#define SKEL_MINB {os.environ['LM_MINB']}\n" + LMOSEM_LANES
    LMOSEM_LANES_PREPARED = f"#define SKEL_MINB {os.environ['LM_MINB']}\n" + LMOSEM_LANES_PREPARED
ev = si.lmosem_events(1_000_000, subset=0)
Ds = [int(x) for x in os.environ.get("LM_DS", "1,2,4,8").split(",")]
LANES = [int(x) for x in os.environ.get("LM_LANES", "1,2,4,8,16").split(",")]
BLOCKS = [int(x) for x in os.environ.get("LM_BLOCKS", "128,256").split(",")]
with skel.Context(1) as ctx:
    stream = torch.cuda.ExternalStream(ctx.stream(0))
    f = ctx.vector(n=150 * 150 * 280, dtype=np.float32).fill(np.float32(1))
    c = ctx.vector(n=150 * 150 * 280, dtype=np.float32)
    dims = [np.int32(150), np.int32(150), np.int32(280)]

    def timed(fn, reps=20):
        for _ in range(3):
            fn()
        ctx.sync()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(stream)
        for _ in range(reps):
            fn()
        e1.record(stream)
        ctx.sync()
        return e0.elapsed_time(e1) / reps

    for D in Ds:
        part = ev[: 1_000_000 // D]
        for order in ("given", "length"):
            e = ctx.vector(part)
            if order == "length":  # ordered on the device (lmosem.LMOSEM.order_on_device)
                e = LMOSEM(ctx, order="device").order_on_device(e)
            for blk in BLOCKS:
                ctx.set_block_size(blk)
                res = {"D": D, "events": len(part), "order": order, "block": blk}
                src1 = LMOSEM_ERROR if order == "given" else LMOSEM_ERROR_PREPARED
                res["map_ms"] = round(timed(lambda: ctx.map(src1, e, None, args=[f, c, *dims])), 4)
                srcl = LMOSEM_LANES if order == "given" else LMOSEM_LANES_PREPARED
                for L in LANES:
                    res[f"lanes{L}_ms"] = round(timed(lambda: ctx.map_lanes(srcl, e, None, L, args=[f, c, *dims])), 4)
                print(json.dumps(res), flush=True)
            ctx.set_block_size(0)
            e.destroy()
