"""Small end-to-end exercise of every kernel family, for compute-sanitizer.

    compute-sanitizer --tool memcheck|racecheck|synccheck|initcheck python tools/sanitize_run.py

Covers: Map/Zip (aligned 128-bit path and unaligned views), Reduce (TMA ring
and direct path, multi-CTA ordered fold), Scan (persistent look-back, TMA and
direct, several slices), copy/block/single exchanges with combine, the fused
zip_combine, a CUDA graph replay, Mandelbrot and one small LM OSEM subset.
Every result is checked (cheaply, against numpy) so a sanitizer run also
proves the instrumented kernels still compute the right thing.
"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402

import skel_inputs as si  # noqa: E402
from paper_conf_ipps_steuwerkg11_b200 import skel  # noqa: E402
from paper_conf_ipps_steuwerkg11_b200.lmosem import LMOSEM  # noqa: E402
from paper_conf_ipps_steuwerkg11_b200.workloads import MANDELBROT, SAXPY_F32, SUM_F32, SUM_I32  # noqa: E402

N = int(os.environ.get("SAN_N", 300_017))


def check(c, what):
    if not c:
        raise SystemExit(f"FAILED: {what}")
    print("ok", what, flush=True)


with skel.Context(1) as ctx:
    x = si.uniform_int01(N, 1)
    v = ctx.vector(x)
    check(int(ctx.reduce(SUM_I32, v)) == int(x.sum()), "reduce i32")
    out = ctx.vector(n=N, dtype=np.int32)
    ctx.scan(SUM_I32, v, out, np.int32(0))
    check(np.array_equal(out.download(), np.concatenate([[0], np.cumsum(x)[:-1]]).astype(np.int32)), "scan i32")
    f = si.uniform_f32(N, 2)
    vf = ctx.vector(f)
    r = float(ctx.reduce(SUM_F32, vf))
    check(abs(r - float(np.sum(f, dtype=np.float64))) < 1e-4 * float(np.abs(f).sum()), "reduce f32")
    z = ctx.vector(n=N, dtype=np.float32)
    ctx.zip(SAXPY_F32, vf, vf, z, args=[np.float32(2.0)])
    check(np.array_equal(z.download(), (np.float32(2.0) * f + f).astype(np.float32)), "zip saxpy")
    # 12-byte elements: direct (non-TMA) reduce/scan path
    aff = "struct Aff { unsigned a, b, n; };\n" \
          "Aff comp(Aff f, Aff g) { Aff r; r.a = f.a * g.a; r.b = f.b * g.a + g.b; r.n = f.n + g.n; return r; }"
    dt = np.dtype([("a", np.uint32), ("b", np.uint32), ("n", np.uint32)])
    m = np.zeros(5000, dt)
    m["a"], m["b"], m["n"] = 1, np.arange(5000) % 7, 1
    rr = ctx.reduce(aff, ctx.vector(m))
    check(int(rr["n"]) == 5000 and int(rr["b"]) == int((np.arange(5000) % 7).sum()), "reduce 12-byte")
    ident = np.zeros(1, dt)
    ident["a"] = 1
    so = ctx.vector(n=5000, dtype=dt)
    ctx.scan(aff, ctx.vector(m), so, ident[0])
    check(int(so.download()["n"][-1]) == 4999, "scan 12-byte")
    # graph replay of a Map + Reduce_to step
    acc = ctx.vector(n=1, dtype=np.float32)
    ctx.map("float sq(float v){ return v * v; }", vf, z)
    ctx.reduce_to(SUM_F32, z, acc)
    g = ctx.capture(lambda: (ctx.map("float sq(float v){ return v * v; }", vf, z), ctx.reduce_to(SUM_F32, z, acc)))
    g.launch()
    check(abs(float(acc.download()[0]) - float((f.astype(np.float64) ** 2).sum())) < 1e-3 * N, "graph replay")
    # Mandelbrot and one LM OSEM subset (small)
    pos = si.mandelbrot_positions(256, 192)
    mo = ctx.vector(n=pos.size, dtype=np.int32)
    ctx.map(MANDELBROT, ctx.vector(pos), mo, args=[np.int32(64)])
    check(int(mo.download().max()) == 64, "mandelbrot")
    ev = si.lmosem_events(2000, subset=0)
    rec = LMOSEM(ctx)
    rec.subset(rec.events(ev))
    img = rec.image()
    check(np.isfinite(img).all() and int((img != 1.0).sum()) > 1000, "lmosem subset")
    # round 2: lanes Map (LM OSEM pieces), on-device ordering + shared-memory staged
    # 24-byte Map, persistent Scan (cooperative) at a size above the small path
    recd = LMOSEM(ctx, order="device", lanes=4)
    recd.subset(recd.events(ev))
    img2 = recd.image()
    check(float(np.abs(img2 - img).max()) < 1e-3, "lmosem lanes + device order")
    from paper_conf_ipps_steuwerkg11_b200.workloads import (MANDELBROT_PAIRS, MANDELBROT_PERIODIC,  # noqa: E402
                                                            MANDELBROT_TILES)
    pos2 = pos.view(si.POS2_DTYPE)
    mp = ctx.vector(n=pos2.size, dtype=si.CNT2_DTYPE)
    ctx.map(MANDELBROT_PAIRS, ctx.vector(pos2), mp, args=[np.int32(64)])
    check(np.array_equal(mp.download().view(np.int32), mo.download()), "mandelbrot pairs")
    ctx.map(MANDELBROT_PERIODIC, ctx.vector(pos), mo, args=[np.int32(64)])
    img_t = ctx.vector(n=pos.size, dtype=np.int32)
    ctx.map_index(MANDELBROT_TILES, pos.size, None, args=[img_t, np.int32(256), np.int32(192), np.int32(64)])
    img_t.mark_device_modified()
    check(np.array_equal(img_t.download(), mo.download()), "mandelbrot periodic + tiles")
    big = si.uniform_int01(1 << 22, 5)
    bo = ctx.vector(n=big.size, dtype=np.int32)
    ctx.scan(SUM_I32, ctx.vector(big), bo, np.int32(0))
    check(int(bo.download()[-1]) == int(big[:-1].sum()), "persistent scan (cooperative)")

with skel.Context(3) as ctx:  # virtual devices: exchanges, unaligned views, fused zip_combine
    x = si.uniform_int01(N, 3)
    v = ctx.vector(x)
    v.set_distribution(skel.COPY)
    w = ctx.vector(n=N, dtype=np.int32)
    ctx.map("int id(int a){ return a; }", v, w)
    w.set_distribution(skel.BLOCK)  # aliased, unaligned parts
    check(int(ctx.reduce(SUM_I32, w)) == int(x.sum()), "reduce on unaligned views")
    so = ctx.vector(n=N, dtype=np.int32)
    ctx.scan(SUM_I32, w, so, np.int32(0))
    check(int(so.download()[-1]) == int(x[:-1].sum()), "scan across devices")
    w.set_distribution(skel.COPY)
    w.set_distribution(skel.BLOCK, skel.COMBINE_ADD)
    check(np.array_equal(w.download(), 3 * x), "copy->block add")
    ev = si.lmosem_events(3000, subset=0)
    rec = LMOSEM(ctx)
    rec.subset(rec.events(ev), fused=True)
    img = rec.image()
    check(np.isfinite(img).all() and int((img != 1.0).sum()) > 1000, "fused zip_combine")
    from paper_conf_ipps_steuwerkg11_b200.mandelbrot import CyclicMandelbrot  # noqa: E402
    cyc = CyclicMandelbrot(ctx, 256, 190).counts(64)
    check(int(cyc.max()) == 64 and cyc.size == 256 * 190, "cyclic rows (gather + un-permute)")
print("sanitize_run: all ok")
