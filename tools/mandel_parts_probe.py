"""Where the Mandelbrot Map's time goes at 4096x3072: the same functions on
(a) the paper image, (b) an all-member image (every c = -0.1+0.1i: 256 updates
per pixel, no divergence -- the steady block loop alone), (c) an all-escape
image (every c = 3: one update per pixel -- the per-pixel overhead alone).
Prints one JSON line; `ideal_us` is 8 FP32 ops per update at the nominal
148 x 128 lanes x 1.965 GHz."""
import json, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import (MANDELBROT, MANDELBROT_BLOCKED, MANDELBROT_PAIRS,
                                                        MANDELBROT_PERIODIC, MANDELBROT_PAIRS_PERIODIC)
extra = {}
for kv in os.environ.get("MANDEL_EXTRA", "").split(";"):
    if "=" in kv:
        k, v = kv.split("=", 1)
        extra[k] = open(v).read() if os.path.exists(v) else v

W, H = int(os.environ.get("MANDEL_W", "4096")), int(os.environ.get("MANDEL_H", "3072"))
cap = int(os.environ.get("MANDEL_CAP", "256"))
peak = 148 * 128 * 1.965e9
paper = si.mandelbrot_positions(W, H)
members = np.zeros_like(paper)
members["re"], members["im"] = -0.1, 0.1
escape = np.zeros_like(paper)
escape["re"], escape["im"] = 3.0, 0.0
res = {"cap": cap}
with skel.Context(1) as ctx:
    st = torch.cuda.ExternalStream(ctx.stream(0))

    def timed(fn, n=10):
        for _ in range(3):
            fn()
        ctx.sync()
        g = ctx.capture(fn)
        g.launch()
        ctx.sync()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(st)
        for _ in range(n):
            g.launch()
        e1.record(st)
        ctx.sync()
        g.destroy()
        return e0.elapsed_time(e1) / n

    fns = {"paper": MANDELBROT, "blocked": MANDELBROT_BLOCKED, "pairs": MANDELBROT_PAIRS,
           "periodic": MANDELBROT_PERIODIC, "pairs_periodic": MANDELBROT_PAIRS_PERIODIC}
    here = os.path.dirname(os.path.abspath(__file__))
    if os.environ.get("MANDEL_DYN"):
        fns["dyn_blocked"] = MANDELBROT_BLOCKED + open(os.path.join(here, "mandel_dyn_exp.cu")).read()
    MX = "#define MANDEL_MAXTEST 1\n"
    fns.update({"blocked_max": MX + MANDELBROT_BLOCKED, "periodic_max": MX + MANDELBROT_PERIODIC,
                "periodic_max16": MX + "#define MANDEL_B 16\n" + MANDELBROT_PERIODIC,
                "nr": "#define MANDEL_NOREPLAY 1\n" + MANDELBROT_BLOCKED,
                "nr_periodic": "#define MANDEL_NOREPLAY 1\n#define MANDEL_PERIODIC 1\n" + MANDELBROT_BLOCKED,
                "nr_periodic_pre4": "#define MANDEL_NOREPLAY 1\n#define MANDEL_PERIODIC 1\n#define MANDEL_PRE 4\n" + MANDELBROT_BLOCKED,
                "nr_periodic_b4": "#define MANDEL_NOREPLAY 1\n#define MANDEL_PERIODIC 1\n#define MANDEL_B 4\n" + MANDELBROT_BLOCKED,
                "p2_max": MX + "#define MANDEL_PERIODIC 2\n#define MANDEL_PRE 8\n" + MANDELBROT_BLOCKED,
                "p2_max_b16": MX + "#define MANDEL_PERIODIC 2\n#define MANDEL_PRE 8\n#define MANDEL_B 16\n" + MANDELBROT_BLOCKED,
                "p2_max_b4": MX + "#define MANDEL_PERIODIC 2\n#define MANDEL_PRE 8\n#define MANDEL_B 4\n" + MANDELBROT_BLOCKED,
                "pairs_nr": "#define MANDEL_NOREPLAY 1\n" + MANDELBROT_PAIRS,
                "pairs_nr_periodic": "#define MANDEL_NOREPLAY 1\n" + MANDELBROT_PAIRS_PERIODIC,
                "pairs_nr_periodic_p4": "#define MANDEL_NOREPLAY 1\n#define MANDEL_P 4\n" + MANDELBROT_PAIRS_PERIODIC,
                "pairs_nr_periodic_p0": "#define MANDEL_NOREPLAY 1\n#define MANDEL_P 0\n" + MANDELBROT_PAIRS_PERIODIC,
                "pairs_nrf_periodic": "#define MANDEL_NOREPLAY 1\n#define MANDEL_NR_FSETP 1\n" + MANDELBROT_PAIRS_PERIODIC,
                "pairs_nrf_periodic_pb16": "#define MANDEL_NOREPLAY 1\n#define MANDEL_NR_FSETP 1\n#define MANDEL_PB 16\n" + MANDELBROT_PAIRS_PERIODIC,
                "pairs_nrf_periodic_pb4": "#define MANDEL_NOREPLAY 1\n#define MANDEL_NR_FSETP 1\n#define MANDEL_PB 4\n" + MANDELBROT_PAIRS_PERIODIC,
                "pairs_periodic_minb12": "#define SKEL_MINB 12\n" + MANDELBROT_PAIRS_PERIODIC,
                "pairs_periodic_minb16": "#define SKEL_MINB 16\n" + MANDELBROT_PAIRS_PERIODIC,
                "periodic_minb16": "#define SKEL_MINB 16\n" + MANDELBROT_PERIODIC,
                "periodic_g15": "#define MANDEL_SAVE_NEXT(s) ((s) + ((s) >> 1) + ((s) < 2))\n" + MANDELBROT_PERIODIC,
                "periodic_g125": "#define MANDEL_SAVE_NEXT(s) ((s) + ((s) >> 2) + ((s) < 4))\n" + MANDELBROT_PERIODIC,
                "pairs_periodic_g15": "#define MANDEL_SAVE_NEXT(s) ((s) + ((s) >> 1) + ((s) < 2))\n" + MANDELBROT_PAIRS_PERIODIC,
                "pairs_periodic_g125": "#define MANDEL_SAVE_NEXT(s) ((s) + ((s) >> 2) + ((s) < 4))\n" + MANDELBROT_PAIRS_PERIODIC,
                "periodic_g3": "#define MANDEL_SAVE_NEXT(s) ((s) * 3)\n" + MANDELBROT_PERIODIC,
                "periodic_g4": "#define MANDEL_SAVE_NEXT(s) ((s) << 2)\n" + MANDELBROT_PERIODIC,
                "pairs_periodic_g3": "#define MANDEL_SAVE_NEXT(s) ((s) * 3)\n" + MANDELBROT_PAIRS_PERIODIC,
                "pairs_periodic_g4": "#define MANDEL_SAVE_NEXT(s) ((s) << 2)\n" + MANDELBROT_PAIRS_PERIODIC,
                "pairs_max": MX + MANDELBROT_PAIRS, "pairs_periodic_max": MX + MANDELBROT_PAIRS_PERIODIC})
    rf = open(os.path.join(here, "mandel_refill_exp.cu")).read()
    for P in (64, 128, 256, 512, 1024):
        fns[f"refill_{P}"] = f"#define MR_P {P}\n" + rf
    fns.update(extra)
    if os.environ.get("MANDEL_ONLY"):
        keep = os.environ["MANDEL_ONLY"].split(",")
        fns = {k: v for k, v in fns.items() if k in keep}
    images = (("paper", paper), ("members", members), ("escape", escape))
    if os.environ.get("MANDEL_IMAGES"):
        images = tuple(im for im in images if im[0] in os.environ["MANDEL_IMAGES"].split(","))
    if os.environ.get("MANDEL_BLOCK"):
        ctx.set_block_size(int(os.environ["MANDEL_BLOCK"]))
    for img_name, pos in images:
        vin = ctx.vector(pos)
        vin2 = ctx.vector(pos.view(si.POS2_DTYPE))
        row = {}
        counts = None
        for name, src in fns.items():
            two = "pairs" in name or "PAIRS" in name[:0]
            two = two or src.find("Pos2 c") >= 0
            v = vin2 if two else vin
            out = ctx.vector(n=v.n, dtype=si.CNT2_DTYPE if two else np.int32)
            if name.startswith("refill"):
                P = int(name.split("_")[1]) if "_" in name else 256
                npix = vin.n
                nthr = -(-npix // P) * 32
                img = ctx.vector(n=npix, dtype=np.int32)
                rargs = [img, np.uint32(npix), np.int32(W), np.int32(H), np.int32(cap)]
                srcr = src
                ms = timed(lambda: ctx.map_index(srcr, nthr, None, args=rargs))
                img.mark_device_modified()
                out.upload(img.download())
                img.destroy()
            elif name.startswith("dyn"):
                nthr = 148 * 2048
                ctr = ctx.vector(np.zeros(2, np.uint32))
                img = ctx.vector(n=vin.n, dtype=np.int32)
                dargs = [vin, img, ctr, np.uint32(vin.n), np.uint32(nthr // 32), np.int32(cap)]
                ms = timed(lambda: ctx.map_index(src, nthr, None, args=dargs))
                img.mark_device_modified()
                out.upload(img.download())
                ctr.destroy()
                img.destroy()
            else:
                ms = timed(lambda: ctx.map(src, v, out, args=[np.int32(cap)]))
            got = out.download().view(np.int32)
            if counts is None:
                counts = got
            row[name] = {"us": round(ms * 1e3, 1), "same": bool(np.array_equal(got, counts))}
            out.destroy()
        iters = int(counts.astype(np.int64).sum())
        row["sum_iter"] = iters
        row["ideal_us"] = round(8 * iters / peak * 1e6, 1)
        res[img_name] = row
        vin.destroy()
        vin2.destroy()
print(json.dumps(res))
