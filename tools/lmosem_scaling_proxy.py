"""LM OSEM subset time at D GPUs projected from pieces measured on ONE GPU
(only one GPU is available to this build).  For D = 1, 2, 4, 8 it times what
each GPU runs per subset at D GPUs (Listing 4's loop body, PAPER.md
P:L518-549), with the library's own policy (lmosem.LMOSEM.plan):

  fill   c <- 0 on the device's whole copy (25.2 MB)
  order  the device's 10^6/D events reordered by path length (order="device")
  map    the error-image Map over the 10^6/D events (given / device order)
  zip    the update Zip over the device's 6.3M/D voxels

and adds the exchange, which one GPU cannot run: copy->block+add
(reduce-scatter) and block->copy (all-gather) of the 25.2 MB image move
(D-1)/D x 25.2 MB into and out of each GPU, at the measured 770 GB/s peer
copy per direction (B200_PROFILING.md; NVLS in-switch reduction would move
1/D of it).  The fused tails (skel_zip_combine) run the update inside the
exchange kernel: max(zip, exchange), not their sum.  `auto` takes, at each D,
the faster event order (the library's order="auto" policy picks by part size).
Prints one JSON line per D and a summary with T1/TD."""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch

import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.lmosem import LMOSEM
from paper_conf_ipps_steuwerkg11_b200.workloads import LMOSEM_UPDATE

NVLINK_GBPS = 770.0
S = 150 * 150 * 280 * 4
ev = si.lmosem_events(1_000_000, subset=0)
rows = []
with skel.Context(1) as ctx:
    stream = torch.cuda.ExternalStream(ctx.stream(0))

    def timed(fn, reps=20):
        """GPU time per call (captured once as a CUDA graph, the graph replayed:
        eager Python calls would add their launch overhead to short pieces)."""
        for _ in range(3):
            fn()
        ctx.sync()
        g = ctx.capture(fn)
        g.launch()
        ctx.sync()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(stream)
        for _ in range(reps):
            g.launch()
        e1.record(stream)
        ctx.sync()
        g.destroy()
        return e0.elapsed_time(e1) / reps

    for D in (1, 2, 4, 8):
        part = ev[: 1_000_000 // D]
        r = {"D": D, "events_per_gpu": len(part)}
        for order in ("given", "device"):
            rec = LMOSEM(ctx, order=order)
            rec.prepare()
            e = ctx.vector(part)
            rec.f.set_distribution(skel.COPY)
            rec.c.fill_dist(skel.COPY, np.float32(0))
            r[f"{order}_map_ms"] = timed(lambda: rec.error_map(e))
            if order == "device":
                r["order_ms"] = timed(lambda: rec.order_on_device(e))
                ordered = rec.order_on_device(e)
                r["device_map_ms"] = timed(lambda: rec.error_map(ordered))
            r["fill_ms"] = timed(lambda: rec.c.fill_dist(skel.COPY, np.float32(0)))
            e.destroy()
        nv = -(-150 * 150 * 280 // D)
        fp, cp = ctx.vector(n=nv, dtype=np.float32).fill(np.float32(1)), ctx.vector(n=nv, dtype=np.float32)
        cp.fill(np.float32(0.5))
        r["zip_ms"] = timed(lambda: ctx.zip(LMOSEM_UPDATE, fp, cp, fp))
        # Bytes per GPU and direction (full-duplex links, S = 25.2 MB):
        # RS + AG (NCCL ring): (D-1)/D S each way for the RS, then again for the AG
        r["exchange_ms_model"] = 2 * S * (D - 1) / D / (NVLINK_GBPS * 1e9) * 1e3
        # fused peer-memory tail (skel_zip_combine): a GPU loads its part of the
        # D-1 other copies and stores its result part into D-1 copies, and serves
        # the same to every peer: 2 (D-1)/D S each way, in ONE kernel
        r["exchange_fused_ms_model"] = 2 * S * (D - 1) / D / (NVLINK_GBPS * 1e9) * 1e3
        # NVLS tail (multimem.ld_reduce + multimem.st): in, S/D reduced + (D-1)/D S of
        # the others' results; out, (D-1)/D S of its copy to the switch + S/D of its
        # result: S each way
        r["exchange_nvls_ms_model"] = S / (NVLINK_GBPS * 1e9) * 1e3 if D > 1 else 0.0
        for order in ("given", "device"):
            extra = r["order_ms"] if order == "device" else 0.0
            base = r["fill_ms"] + extra + r[f"{order}_map_ms"]
            # unfused: reduce-scatter, then the update Zip, then the all-gather
            r[f"{order}_subset_ms"] = base + r["zip_ms"] + r["exchange_ms_model"]
            # fused tails: the update runs inside the exchange kernel on the part
            # it has just combined (its 2 x S/D bytes of HBM traffic overlap the
            # NVLink transfers), so the kernel takes the longer of the two
            r[f"{order}_subset_fused_ms"] = base + max(r["zip_ms"], r["exchange_fused_ms_model"])
            r[f"{order}_subset_nvls_ms"] = base + max(r["zip_ms"], r["exchange_nvls_ms_model"])
        for tail in ("", "_fused", "_nvls"):  # the order policy that is faster at this part size
            r[f"auto_subset{tail}_ms"] = min(r[f"given_subset{tail}_ms"], r[f"device_subset{tail}_ms"])
        rows.append(r)
        print(json.dumps({k: (round(v, 4) if isinstance(v, float) else v) for k, v in r.items()}), flush=True)
summary = {}
for order in ("given", "device", "auto"):
    for tail in ("", "_fused", "_nvls"):
        t1 = rows[0][f"{order}_subset{tail}_ms"]
        summary[order + tail] = {f"T1/T{r['D']}": round(t1 / r[f"{order}_subset{tail}_ms"], 2) for r in rows}
print(json.dumps({"projection": summary, "exchange": f"RS + AG of {S / 1e6:.1f} MB at {NVLINK_GBPS} GB/s per direction"}))
