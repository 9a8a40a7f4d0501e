"""Feasibility probe: does a SPATIAL order of the LM OSEM events (warps of
nearly parallel, adjacent lines of response) speed up the error-image Map?
Events are sorted on the host here (numpy) by different keys and the Map timed
in each order (one thread per event with 16-byte forward gathers, and the
4-lane Map), at 10^6 events (one GPU) and 1.25*10^5 (one GPU's part at 8).
Prints one JSON line per (events, order)."""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch

import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import (LMOSEM_ERROR, LMOSEM_ERROR_PREPARED, LMOSEM_LANES,
                                                        LMOSEM_LANES_PREPARED)

ev_all = si.lmosem_events(1_000_000, subset=0)


def keys(ev, nphi, ns, nz, nt):
    x1, y1, z1 = (ev[k].astype(np.float64) for k in ("x1", "y1", "z1"))
    x2, y2, z2 = (ev[k].astype(np.float64) for k in ("x2", "y2", "z2"))
    dx, dy, dz = x2 - x1, y2 - y1, z2 - z1
    r = np.sqrt(dx * dx + dy * dy)
    phi = np.mod(np.arctan2(dy, dx), 2 * np.pi)
    s = ((x1 - 75.0) * dy - (y1 - 75.0) * dx) / r
    zm = 0.5 * (z1 + z2)
    t = dz / r
    b_phi = np.minimum((phi / (2 * np.pi) * nphi).astype(np.int64), nphi - 1)
    b_s = np.clip(((s + 110.0) / 220.0 * ns).astype(np.int64), 0, ns - 1)
    b_z = np.clip((zm / 280.0 * nz).astype(np.int64), 0, nz - 1)
    b_t = np.clip(((t + 0.32) / 0.64 * nt).astype(np.int64), 0, nt - 1)
    return ((b_phi * ns + b_s) * nz + b_z) * nt + b_t


def length_key(ev):
    d = np.abs(ev["x2"].astype(np.float64) - ev["x1"]) + np.abs(ev["y2"].astype(np.float64) - ev["y1"]) + \
        np.abs(ev["z2"].astype(np.float64) - ev["z1"])
    return -d


with skel.Context(1) as ctx:
    st = torch.cuda.ExternalStream(ctx.stream(0))
    f = ctx.vector(n=150 * 150 * 280, dtype=np.float32).fill(np.float32(1))
    c = ctx.vector(n=150 * 150 * 280, dtype=np.float32)
    dims = [np.int32(150), np.int32(150), np.int32(280)]

    def timed(fn, reps=10):
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
        return round(e0.elapsed_time(e1) / reps, 4)

    ctx.set_block_size(128)
    for n in (1_000_000, 125_000):
        ev = ev_all[:n]
        orders = {"given": np.arange(n), "length": np.argsort(length_key(ev), kind="stable")}
        for cfg in ((64, 64, 8, 4), (128, 128, 8, 2), (64, 128, 16, 2), (256, 64, 4, 2), (32, 256, 8, 2)):
            orders["spatial_%d_%d_%d_%d" % cfg] = np.argsort(keys(ev, *cfg), kind="stable")
        for name, idx in orders.items():
            e = ctx.vector(np.ascontiguousarray(ev[idx]))
            res = {"events": n, "order": name}
            res["map1_prepared_ms"] = timed(lambda: ctx.map(LMOSEM_ERROR_PREPARED, e, None, args=[f, c, *dims]))
            res["map1_given_fn_ms"] = timed(lambda: ctx.map(LMOSEM_ERROR, e, None, args=[f, c, *dims]))
            res["lanes4_prepared_ms"] = timed(lambda: ctx.map_lanes(LMOSEM_LANES_PREPARED, e, None, 4, args=[f, c, *dims]))
            res["lanes4_given_fn_ms"] = timed(lambda: ctx.map_lanes(LMOSEM_LANES, e, None, 4, args=[f, c, *dims]))
            print(json.dumps(res), flush=True)
            e.destroy()
