"""Pieces of the on-device LM OSEM event ordering (workloads/lmosem_order.cu),
timed one by one at 10^6 events: the key alone, the key + atomics with and
without warp aggregation, and the scatter."""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch

import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import (LMOSEM_ERROR, LMOSEM_ORDER_HIST, LMOSEM_ORDER_SCATTER,
                                                        LMOSEM_ORDER_SLOTS, source)

ORD = LMOSEM_ERROR + source("lmosem_order")
KEY = ORD + "\nint lm_key(Event e, int nx, int ny, int nz, int nb) { return lm_slot(e, nx, ny, nz, nb); }\n"
BUCKET = ORD + "\nint lm_key(Event e, int nx, int ny, int nz, int nb) { return lm_bucket(e, nx, ny, nz, nb); }\n"
COPY = ORD + "\nint lm_key(Event e, int nx, int ny, int nz, int nb) { return __float_as_int(e.x1) ^ nb; }\n"
HIST_PLAIN = ORD + """
void lm_h(Event e, int *hist, int nx, int ny, int nz, int nb) { atomicAdd(&hist[lm_slot(e, nx, ny, nz, nb)], 1); }
"""
ev = si.lmosem_events(1_000_000, subset=0)
with skel.Context(1) as ctx:
    st = torch.cuda.ExternalStream(ctx.stream(0))
    e = ctx.vector(ev)
    key = ctx.vector(n=ev.size, dtype=np.int32)
    hist = ctx.vector(n=LMOSEM_ORDER_SLOTS, dtype=np.int32).fill(np.int32(0))
    out = ctx.vector(n=ev.size, dtype=ev.dtype)
    dims = [np.int32(150), np.int32(150), np.int32(280), np.int32(64)]

    def timed(fn, reps=20):
        """GPU time per call: the calls are captured once as a CUDA graph and the
        graph replayed (eager timing would measure the Python/ctypes launch rate)."""
        for _ in range(3):
            fn()
        ctx.sync()
        g = ctx.capture(fn)
        g.launch()
        ctx.sync()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(st)
        for _ in range(reps):
            g.launch()
        e1.record(st)
        ctx.sync()
        g.destroy()
        return round(e0.elapsed_time(e1) / reps * 1e3, 2)
    res = {}
    for blk in (256, 128):
        ctx.set_block_size(blk)
        res[f"copy_key_us_{blk}"] = timed(lambda: ctx.map(COPY, e, key, args=dims))
        res[f"bucket_key_us_{blk}"] = timed(lambda: ctx.map(BUCKET, e, key, args=dims))
        res[f"slot_key_us_{blk}"] = timed(lambda: ctx.map(KEY, e, key, args=dims))
        res[f"hist_match_us_{blk}"] = timed(lambda: ctx.map(LMOSEM_ORDER_HIST, e, None, args=[hist, *dims]))
        res[f"hist_plain_us_{blk}"] = timed(lambda: ctx.map(HIST_PLAIN, e, None, args=[hist, *dims]))
        hist.fill(np.int32(0))
        res[f"scatter_us_{blk}"] = timed(lambda: (hist.fill(np.int32(0)),
                                                  ctx.map(LMOSEM_ORDER_SCATTER, e, None, args=[hist, out, *dims])))
        from paper_conf_ipps_steuwerkg11_b200.lmosem import LMOSEM
        rec = LMOSEM(ctx, order="device")
        rec.prepare()
        res[f"order_on_device_us_{blk}"] = timed(lambda: rec.order_on_device(e))
    ctx.set_block_size(0)
    print(json.dumps(res))
