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
from .workloads import LMOSEM_ERROR, LMOSEM_UPDATE

DIMS = (150, 150, 280)


class LMOSEM:
    def __init__(self, ctx: skel.Context, dims=DIMS, f0: float = 1.0):
        self.ctx = ctx
        self.dims = tuple(int(d) for d in dims)
        self.nvox = int(np.prod(self.dims))
        self.f = ctx.vector(n=self.nvox, dtype=np.float32)
        self.c = ctx.vector(n=self.nvox, dtype=np.float32)
        self.f.fill_dist(skel.BLOCK, np.float32(f0))  # f0 = 1 everywhere (reading R10(ii))
        self.dims_args = [np.int32(d) for d in self.dims]

    def prepare(self):
        self.ctx.prepare("map", LMOSEM_ERROR)
        self.ctx.prepare("zip", LMOSEM_UPDATE)

    def events(self, ev: np.ndarray) -> skel.Vector:
        """Vector<Event> of one subset, block-distributed (Listing 4)."""
        v = self.ctx.vector(ev)
        v.set_distribution(skel.BLOCK)
        return v

    def subset(self, events: skel.Vector, fused: bool = False):
        """One iteration of Listing 4's loop body.  fused=True runs the tail
        (combine c, update f, redistribute f) as one peer-memory kernel."""
        ctx, f, c = self.ctx, self.f, self.c
        f.set_distribution(skel.COPY)                     # block -> copy: all-gather (no-op after a fused tail)
        c.fill_dist(skel.COPY, np.float32(0))             # fresh zero copy on every device
        ctx.map(LMOSEM_ERROR, events, None, args=[f, c, *self.dims_args])
        c.mark_device_modified()                          # dataOnDevicesModified()
        if fused:
            ctx.zip_combine(LMOSEM_UPDATE, f, c, skel.COMBINE_ADD, f)
            return
        f.set_distribution(skel.BLOCK)                    # copy -> block: local slice
        c.set_distribution(skel.BLOCK, skel.COMBINE_ADD)  # copy -> block + add: reduce-scatter
        ctx.zip(LMOSEM_UPDATE, f, c, f)                   # f[j] *= c[j] where c[j] > 0

    def image(self) -> np.ndarray:
        return self.f.download()
