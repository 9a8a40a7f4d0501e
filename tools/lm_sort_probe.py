import os, sys
sys.path.insert(0, os.getcwd())
import numpy as np, torch
import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import LMOSEM_ERROR, LMOSEM_VISITS
ev = si.lmosem_events(1_000_000, subset=0)
with skel.Context(1) as ctx:
    st = torch.cuda.ExternalStream(ctx.stream(0))
    f = ctx.vector(n=150*150*280, dtype=np.float32).fill(np.float32(1))
    c = ctx.vector(n=150*150*280, dtype=np.float32)
    dims = [np.int32(150), np.int32(150), np.int32(280)]
    e = ctx.vector(ev)
    nv = ctx.vector(n=len(ev), dtype=np.int32)
    ctx.map(LMOSEM_VISITS, e, nv, args=dims)
    L = nv.download()
    orders = {"given": np.arange(len(ev)), "sorted": np.argsort(L, kind="stable"),
              "sorted_desc": np.argsort(-L, kind="stable")}
    # 8-way interleave of the sorted order (what each of 8 GPUs would get in a block part)
    s = np.argsort(L, kind="stable"); D = 8
    orders["sorted_dealt8"] = np.concatenate([s[k::D] for k in range(D)])
    for name, o in orders.items():
        ee = ctx.vector(ev[o])
        for D in (1, 8):
            n = len(ev) // D
            sub = ctx.vector(ev[o][:n]) if D > 1 else ee
            for _ in range(3): ctx.map(LMOSEM_ERROR, sub, None, args=[f, c, *dims])
            ctx.sync()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(st)
            for _ in range(10): ctx.map(LMOSEM_ERROR, sub, None, args=[f, c, *dims])
            e1.record(st); ctx.sync()
            print(name, D, round(e0.elapsed_time(e1) / 10, 4), "ms")
