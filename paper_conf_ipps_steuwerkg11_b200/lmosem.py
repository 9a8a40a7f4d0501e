"""List-mode OSEM on the skeletons, structured as Listing 4 of the paper
(P:L518-549): events block-distributed, reconstruction image f and error
image c copy-distributed during the Map, c merged by copy->block+add, and f
updated by a Zip on the blocks.

Reading R10(i): c is reset to 0 at the start of every subset (Listing 3/4 do
not show it, but without it the combine would re-add the previous subset's
error image D times).
"""
from __future__ import annotations

import numpy as np

from . import skel
from .workloads import LMOSEM_ERROR, LMOSEM_ERROR_PREPARED, LMOSEM_UPDATE

DIMS = (150, 150, 280)


def order_by_path(ev: np.ndarray, dims=DIMS) -> np.ndarray:
    """The events of a subset reordered longest path first (host preprocessing,
    like reading the subset from file).  List-mode events carry no
    order, and the error image is a sum over them, so any order gives the same
    image up to float rounding (R10(x)).  With similar path lengths next to each
    other, the 32 rays of a warp finish together (thread efficiency) and the
    longest rays start first (shorter launch tail): DESIGN.md §4.2.
    Key: the L1 length |dx|+|dy|+|dz| of the segment clipped to the volume
    (slab clipping, float64) -- proportional to the voxel steps of the walk."""
    p = np.stack([ev["x1"], ev["y1"], ev["z1"]]).astype(np.float64)
    d = np.stack([ev["x2"], ev["y2"], ev["z2"]]).astype(np.float64) - p
    amin = np.zeros(len(ev))
    amax = np.ones(len(ev))
    for a, n in enumerate(dims):
        nz = d[a] != 0
        with np.errstate(divide="ignore", invalid="ignore"):
            a0 = np.where(nz, (0.0 - p[a]) / d[a], -np.inf)
            a1 = np.where(nz, (float(n) - p[a]) / d[a], np.inf)
        inside = (p[a] >= 0) & (p[a] < n)
        amin = np.maximum(amin, np.where(nz, np.minimum(a0, a1), np.where(inside, -np.inf, np.inf)))
        amax = np.minimum(amax, np.where(nz, np.maximum(a0, a1), np.inf))
    key = np.where(amax > amin, (amax - amin) * np.abs(d).sum(axis=0), 0.0)
    return ev[np.argsort(-key, kind="stable")]


def deal_warps(ev: np.ndarray, block: int = 256, warp: int = 32) -> np.ndarray:
    """Events ordered longest path first (order_by_path), then their groups of
    `warp` consecutive events dealt round-robin to the `block`-thread CTAs of a
    one-event-per-thread launch (snake order): a warp keeps rays of similar
    length, and every CTA gets one group from each length range, so the CTAs
    (and the SMs that host them) carry equal work."""
    o = order_by_path(ev)
    n = len(o)
    ng = -(-n // warp)
    per_cta = block // warp
    ncta = -(-ng // per_cta)
    # group g (in length order) goes to slot g // ncta of a CTA dealt in snake
    # order (0..ncta-1, then ncta-1..0, ...), which evens out the CTAs' sums
    gid = np.arange(ng)
    rnd, pos = gid // ncta, gid % ncta
    cta = np.where(rnd % 2 == 0, pos, ncta - 1 - pos)
    dest = cta * per_cta + rnd
    order = np.argsort(dest, kind="stable")
    idx = (order[:, None] * warp + np.arange(warp)[None, :]).ravel()
    return o[idx[idx < n]]


# events per device below which a launch is well under one wave of the GPU
# (148 SMs x 2048 threads); there 128-thread CTAs and warp-dealt order balance
# the SMs better (measured: better at 1.25e5 events per GPU,
# worse at 2.5e5)
SMALL_PART = 150_000


def prepare_part(ev: np.ndarray, dims=DIMS) -> tuple[np.ndarray, int]:
    """(events, CTA size for the error-image Map) for one device's part of a
    subset: longest path first at the default CTA size, or -- for parts below
    SMALL_PART events -- warp groups dealt over 128-thread CTAs."""
    if len(ev) <= SMALL_PART:
        return deal_warps(ev, block=128), 128
    return order_by_path(ev, dims), 0


class LMOSEM:
    def __init__(self, ctx: skel.Context, dims=DIMS, f0: float = 1.0):
        self.ctx = ctx
        self.dims = tuple(int(d) for d in dims)
        self.nvox = int(np.prod(self.dims))
        self.f = ctx.vector(n=self.nvox, dtype=np.float32)
        self.c = ctx.vector(n=self.nvox, dtype=np.float32)
        self.f.fill_dist(skel.BLOCK, np.float32(f0))  # f0 = 1 everywhere (reading R10(ii))
        self.dims_args = [np.int32(d) for d in self.dims]
        self.map_block = 0  # CTA size of the error-image Map (0 = the context's default)
        self.error_src = LMOSEM_ERROR  # LMOSEM_ERROR_PREPARED for prepared event order

    def prepare(self):
        if self.map_block:
            self.ctx.set_block_size(self.map_block)
        self.ctx.prepare("map", self.error_src)
        if self.map_block:
            self.ctx.set_block_size(0)
        self.ctx.prepare("zip", LMOSEM_UPDATE)

    def events(self, ev: np.ndarray, prepare: bool = False) -> skel.Vector:
        """Vector<Event> of one subset, block-distributed (Listing 4).
        prepare=True: each device's part [k*ceil(n/D), ...) reordered by
        prepare_part (the error-image Map then uses the CTA size it picks).
        In rank mode pass the whole subset on every rank, as for a plain upload."""
        if prepare and len(ev):
            D = self.ctx.D
            ps = -(-len(ev) // D)
            parts = []
            for k in range(D):
                part, blk = prepare_part(ev[k * ps:(k + 1) * ps], self.dims)
                parts.append(part)
                if k == 0:
                    self.map_block = blk
            self.error_src = LMOSEM_ERROR_PREPARED
            ev = np.concatenate(parts)
        v = self.ctx.vector(ev)
        v.set_distribution(skel.BLOCK)
        return v

    def subset(self, events: skel.Vector, fused: bool = False):
        """One iteration of Listing 4's loop body.  fused=True runs the tail
        (combine c, update f, redistribute f) as one peer-memory kernel."""
        ctx, f, c = self.ctx, self.f, self.c
        f.set_distribution(skel.COPY)                     # block -> copy: all-gather (no-op after a fused tail)
        c.fill_dist(skel.COPY, np.float32(0))             # fresh zero copy on every device
        if self.map_block:
            ctx.set_block_size(self.map_block)
        ctx.map(self.error_src, events, None, args=[f, c, *self.dims_args])
        if self.map_block:
            ctx.set_block_size(0)
        c.mark_device_modified()                          # dataOnDevicesModified()
        if fused:
            ctx.zip_combine(LMOSEM_UPDATE, f, c, skel.COMBINE_ADD, f)
            return
        f.set_distribution(skel.BLOCK)                    # copy -> block: local slice
        c.set_distribution(skel.BLOCK, skel.COMBINE_ADD)  # copy -> block + add: reduce-scatter
        ctx.zip(LMOSEM_UPDATE, f, c, f)                   # f[j] *= c[j] where c[j] > 0

    def image(self) -> np.ndarray:
        return self.f.download()
