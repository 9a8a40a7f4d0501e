"""Rank-mode (one process per logical device, NCCL) self-test.  Run under
torchrun; every rank uses CUDA device SKEL_TEST_DEVICE (default: its local
rank).  Checks skeleton results and every distribution transition against the
oracle's distribution model; prints one line per rank."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch.distributed as dist

import oracle
import skel_inputs as si
from oracle import distribution as odist
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.lmosem import LMOSEM
from paper_conf_ipps_steuwerkg11_b200.workloads import SUM_F32, SUM_I32

rank, world = int(os.environ["RANK"]), int(os.environ["WORLD_SIZE"])
dev = int(os.environ.get("SKEL_TEST_DEVICE", os.environ.get("LOCAL_RANK", "0")))
dist.init_process_group("gloo")
obj = [skel.unique_id() if rank == 0 else None]
dist.broadcast_object_list(obj, src=0)
fails = []
try:
    ctx = skel.Context(rank=rank, world=world, device=dev, nccl_id=obj[0])
except skel.SkelError as e:
    print(f"rank {rank}: context failed: {e}", flush=True)
    sys.exit(3)


def check(name, ok):
    if not ok:
        fails.append(name)


n = 100_003
x = si.uniform_int01(n, 5)
# reduce / scan across ranks
v = ctx.vector(x)
v.set_distribution(skel.BLOCK)
check("reduce", int(ctx.reduce(SUM_I32, v)) == int(x.sum()))
out = ctx.vector(n=n, dtype=np.int32)
ctx.scan(SUM_I32, v, out, np.int32(0))
check("scan", np.array_equal(out.download(), oracle.skel_scan(SUM_I32, x, 0)))
xf = si.uniform_f32(n, 6)
vf = ctx.vector(xf)
vf.set_distribution(skel.BLOCK)
check("reduce_f32", abs(float(ctx.reduce(SUM_F32, vf)) - oracle.sum_f32_exact(xf)) <= 1e-5 * oracle.abssum_f32(xf))
# every transition
IDENT = "int ident(int x){ return x; }"
for a in (skel.SINGLE, skel.BLOCK, skel.COPY):
    for b in (skel.SINGLE, skel.BLOCK, skel.COPY):
        w0 = ctx.vector(x)
        w0.set_distribution(a)
        w = ctx.vector(n=n, dtype=np.int32)
        ctx.map(IDENT, w0, w)
        w.set_distribution(b)
        check(f"xchg {a}->{b}", np.array_equal(w.download(), x))
# diverged copies combined
mark = "void mark(int i, int* c){ c[i] += 1 + i % 7; }"
for dst in (skel.BLOCK, skel.SINGLE, skel.COPY):
    c = ctx.vector(np.zeros(n, np.int32))
    c.set_distribution(skel.COPY)
    idx = ctx.vector(np.arange(n, dtype=np.int32))
    idx.set_distribution(skel.BLOCK)
    ctx.map(mark, idx, None, args=[c])
    c.mark_device_modified()
    c.set_distribution(dst, skel.COMBINE_ADD)
    want = (1 + np.arange(n) % 7).astype(np.int32)
    for rep in range(int(os.environ.get("SKEL_SELFTEST_REPS", "1"))):
        got = c.download() if rep == 0 else c.download()
        ok = np.array_equal(got, want)
        if not ok:
            bad = np.nonzero(got != want)[0]
            print(f"rank {rank}: combine->{dst} rep {rep}: {bad.size} bad, first {bad[:5]}, got {got[bad[:5]]}, "
                  f"want {want[bad[:5]]}, parts {[c.part(d) for d in range(world)]}", flush=True)
        check(f"combine->{dst}", ok)
# NEXT-2: user-defined combine (gathered on each part's rank, folded in rank order)
MX = "int mx(int a, int b){ return a > b ? a : b; }"
for dst in (skel.BLOCK, skel.SINGLE, skel.COPY):
    base = ((np.arange(n) % 613) - 300).astype(np.int32)
    c = ctx.vector(base)
    c.set_distribution(skel.COPY)
    idx = ctx.vector(np.arange(n, dtype=np.int32))
    idx.set_distribution(skel.BLOCK)
    ctx.map("void mark(int i, int* c){ c[i] = (i * 7919) % 1000 - 500; }", idx, None, args=[c])
    c.mark_device_modified()
    c.set_distribution(dst, MX)
    # rank r's copy: base, with r's block of indices marked; the combine takes the
    # maximum over the ranks' copies (a single rank: its copy, all marked)
    marks = ((np.arange(n) * 7919) % 1000 - 500).astype(np.int32)
    copies = []
    for r in range(world):
        cr = base.copy()
        lo, hi = odist.part_range(n, world, r)
        cr[lo:hi] = marks[lo:hi]
        copies.append(cr)
    want = np.max(np.stack(copies), axis=0)
    check(f"user combine->{dst}", np.array_equal(c.download(), want))
# LM OSEM one subset, then two more with the fused peer-memory tail (CUDA IPC)
ev = si.lmosem_events(20_000, subset=1)
rec = LMOSEM(ctx)
rec.subset(rec.events(ev))
img = rec.image()
want, _, _ = oracle.lmosem_subset(ev, np.ones(150 * 150 * 280))
rel = float(np.linalg.norm(img - want) / np.linalg.norm(want))
check("lmosem", rel <= 1e-4)
subsets = [si.lmosem_events(8_000, subset=l) for l in range(2)]
rec2 = LMOSEM(ctx)
for sub in subsets:
    rec2.subset(rec2.events(sub), fused=True)
want2 = oracle.lmosem_reconstruct(subsets)
rel2 = float(np.linalg.norm(rec2.image() - want2) / np.linalg.norm(want2))
check("lmosem_fused", rel2 <= 1e-4)
print(f"rank {rank}/{world} device {dev}: {'OK' if not fails else 'FAIL ' + ','.join(fails)} (lmosem relL2 {rel:.2e})",
      flush=True)
ctx.close()
dist.destroy_process_group()
sys.exit(1 if fails else 0)
