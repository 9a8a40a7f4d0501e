"""Error-image Map time for one 10^6-event subset under different event orders
(list-mode events carry no order).  Prints ms per Map at D=1 and for the first
1/8 of each order (the per-GPU part at D=8)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch

import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.lmosem import order_by_path
from paper_conf_ipps_steuwerkg11_b200.workloads import LMOSEM_ERROR

ev = si.lmosem_events(1_000_000, subset=0)
p1 = np.stack([ev["x1"], ev["y1"], ev["z1"]]).astype(np.float64)
p2 = np.stack([ev["x2"], ev["y2"], ev["z2"]]).astype(np.float64)
d = p2 - p1
phi = np.mod(np.arctan2(d[1], d[0]), np.pi)                      # LOR angle in the xy-plane
nrm = np.hypot(d[0], d[1])
s = ((p1[0] - 75) * d[1] - (p1[1] - 75) * d[0]) / nrm               # signed distance from the axis
zm = 0.5 * (p1[2] + p2[2])


def sino(phi_bins, s_bins, z_bins):
    k = (np.floor(phi / np.pi * phi_bins).astype(np.int64) * s_bins
         + np.clip(np.floor((s + 110) / 220 * s_bins), 0, s_bins - 1).astype(np.int64)) * z_bins \
        + np.clip(np.floor(zm / 280 * z_bins), 0, z_bins - 1).astype(np.int64)
    return np.argsort(k, kind="stable")


orders = {
    "given": np.arange(len(ev)),
    "length": None,
    "sino_180x220x28": sino(180, 220, 28),
    "sino_360x440x1": sino(360, 440, 1),
    "sino_90x110x56": sino(90, 110, 56),
}
dealt = lambda o: np.concatenate([o[k::8] for k in range(8)])  # noqa: E731
with skel.Context(1) as ctx:
    st = torch.cuda.ExternalStream(ctx.stream(0))
    f = ctx.vector(n=150 * 150 * 280, dtype=np.float32).fill(np.float32(1))
    c = ctx.vector(n=150 * 150 * 280, dtype=np.float32)
    dims = [np.int32(150), np.int32(150), np.int32(280)]
    for name, o in orders.items():
        for D in (1, 8):
            if name == "length":
                part = order_by_path(ev[: len(ev) // D])
            elif D == 1:
                part = ev[o]
            else:  # this GPU's block of a random split, ordered the same way
                blk = np.sort(o[o < len(ev) // D]) if False else None
                sub = ev[: len(ev) // D]
                oo = o[o < len(ev) // D]
                part = sub[oo]
            e = ctx.vector(part)
            for _ in range(7):
                ctx.map(LMOSEM_ERROR, e, None, args=[f, c, *dims])
            ctx.sync()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(st)
            for _ in range(10):
                ctx.map(LMOSEM_ERROR, e, None, args=[f, c, *dims])
            e1.record(st)
            ctx.sync()
            print(name, "D=%d" % D, round(e0.elapsed_time(e1) / 10, 4), "ms", flush=True)
            e.destroy()
