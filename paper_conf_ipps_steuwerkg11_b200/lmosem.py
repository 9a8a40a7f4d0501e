"""List-mode OSEM on the skeletons, structured as Listing 4 of the paper
(P:L518-549): events block-distributed, reconstruction image f and error
image c copy-distributed during the Map, c merged by copy->block+add, and f
updated by a Zip on the blocks.

Reading R10(i): c is reset to 0 at the start of every subset (Listing 3/4 do
not show it, but without it the combine would re-add the previous subset's
error image D times).

The error-image Map (Listing 3 lines 4-13 inside Listing 4's Map) runs in one
of two forms, picked per subset from the events each device holds
(`LMOSEM.plan`):

* a Map with one thread per event (workloads/lmosem_error.cu), or
* a lanes Map (skel_map_lanes) with `lanes` threads per event, each walking an
  alpha piece of the line of response (workloads/lmosem_lanes.cu) -- the form
  that fills the GPU when one device's part of a subset is small (10^6/8
  events at 8 GPUs).

`order="device"` (and `order="auto"`, the default, for parts of at least
AUTO_ORDER_FROM events) first reorders every device's events by path length on
the device with the library's own skeletons (a counting Map, a Scan of the
bucket counts and a scattering Map; workloads/lmosem_order.cu): list-mode
events carry no order and the error image is a sum over events (R10(x)), so
the image is the same up to float rounding, and rays of similar length then
share a warp.
"""
from __future__ import annotations

import numpy as np

from . import skel
from .workloads import (LMOSEM_ERROR, LMOSEM_ERROR_PREPARED, LMOSEM_LANES,
                        LMOSEM_ORDER_BUCKETS, LMOSEM_ORDER_HIST, LMOSEM_ORDER_SCATTER, LMOSEM_ORDER_SLOTS,
                        LMOSEM_UPDATE, SUM_I32)

DIMS = (150, 150, 280)

# CTA size of every error-image Map (measured at 10^6/D events, D = 1..8,
# tools/lm_lanes_probe.py: 128 is as fast or faster than 256 everywhere)
MAP_BLOCK = 128
# events per device from which the one-thread-per-event Map (16-byte forward
# gathers) beats the 4-lane Map (scalar gathers) on length-ordered events
# (round 2, graph replays: 10^6: 1.141 vs 1.147 ms; 5*10^5: 0.589 vs 0.582;
# 2.5*10^5: 0.317 vs 0.300; 1.25*10^5: 0.179 vs 0.160)
ORDERED_LANES_BELOW = 750_000
# order="auto": events per device from which ordering them on the device pays
# for itself (ordering + ordered Map vs the 4-lane Map in the given order:
# 10^6: 0.071 + 1.141 vs 1.287 ms; 2.5*10^5: 0.028 + 0.300 vs 0.335;
# 1.25*10^5: 0.020 + 0.160 vs 0.177)
AUTO_ORDER_FROM = 200_000


class LMOSEM:
    def __init__(self, ctx: skel.Context, dims=DIMS, f0: float = 1.0, order: str = "auto",
                 lanes: int | None = None):
        if order not in ("given", "device", "auto"):
            raise ValueError("order must be 'given', 'device' or 'auto'")
        self.ctx = ctx
        self.dims = tuple(int(d) for d in dims)
        self.nvox = int(np.prod(self.dims))
        self.f = ctx.vector(n=self.nvox, dtype=np.float32)
        self.c = ctx.vector(n=self.nvox, dtype=np.float32)
        self.f.fill_dist(skel.BLOCK, np.float32(f0))  # f0 = 1 everywhere (reading R10(ii))
        self.dims_args = [np.int32(d) for d in self.dims]
        self.order = order
        self.lanes = lanes  # None: LMOSEM.plan decides per subset
        self._hist = self._cursor = self._sorted = None

    # ---- policy ------------------------------------------------------------
    def ordered(self, per_device: int) -> bool:
        """Whether the events are ordered on the device before the Map."""
        return self.order == "device" or (self.order == "auto" and per_device >= AUTO_ORDER_FROM)

    def per_device(self, events: skel.Vector) -> int:
        return -(-events.n // self.ctx.D) if events.distribution == skel.BLOCK else events.n

    def plan(self, per_device: int) -> tuple[str, int]:
        """(error-image function source, lanes) for parts of `per_device`
        events.  Given order: 4 lanes per event at every measured part size
        (10^6/D events, D = 1..8: 1.29 / 0.655 / 0.337 / 0.179 ms against
        1.37 / 0.727 / 0.394 / 0.211 ms with one thread per event).
        Length-ordered events: one thread per event with 16-byte forward
        gathers from ORDERED_LANES_BELOW on, 4 lanes with scalar gathers below
        it (the 16-byte gathers lose once a ray is split into pieces)."""
        ordered = self.ordered(per_device)
        lanes = self.lanes
        if lanes is None:
            lanes = 4 if (not ordered or per_device < ORDERED_LANES_BELOW) else 1
        if lanes == 1:
            return (LMOSEM_ERROR_PREPARED if ordered else LMOSEM_ERROR), 1
        return LMOSEM_LANES, lanes

    def prepare(self):
        """Compile every function a subset may use (before timing or capturing)."""
        ctx = self.ctx
        ctx.set_block_size(MAP_BLOCK)
        for src in (LMOSEM_ERROR, LMOSEM_ERROR_PREPARED):
            ctx.prepare("map", src)
        for src in (LMOSEM_LANES,):
            ctx.prepare("lanes", src)
        ctx.set_block_size(0)
        ctx.prepare("zip", LMOSEM_UPDATE)
        if self.order != "given":
            ctx.prepare("map", LMOSEM_ORDER_HIST)
            ctx.prepare("map", LMOSEM_ORDER_SCATTER)
            ctx.prepare("scan", SUM_I32)

    # ---- data ----------------------------------------------------------------
    def events(self, ev: np.ndarray) -> skel.Vector:
        """Vector<Event> of one subset, block-distributed (Listing 4).
        In rank mode pass the whole subset on every rank, as for a plain upload."""
        v = self.ctx.vector(ev)
        v.set_distribution(skel.BLOCK)
        return v

    def order_on_device(self, events: skel.Vector) -> skel.Vector:
        """Every device's events reordered longest path first, on the device:
        bucket counts (void Map, one atomic per bucket and warp), exclusive Scan
        of the counts, and a void Map that moves each event to its bucket's next
        slot.  Returns a vector with the same distribution and part sizes."""
        ctx, nb = self.ctx, LMOSEM_ORDER_BUCKETS
        if self._hist is None:  # bucket-major counter slots (lmosem_order.cu: lm_slot)
            self._hist = ctx.vector(n=LMOSEM_ORDER_SLOTS, dtype=np.int32)
            self._cursor = ctx.vector(n=LMOSEM_ORDER_SLOTS, dtype=np.int32)
        if self._sorted is None or self._sorted.n != events.n or \
                self._sorted.distribution != events.distribution:
            if self._sorted is not None:
                self._sorted.destroy()
            self._sorted = ctx.vector(n=events.n, dtype=events.dtype)
            self._sorted.fill_dist(events.distribution, np.zeros(1, events.dtype)[0])
        hist, cursor, out = self._hist, self._cursor, self._sorted
        hist.fill_dist(skel.COPY, np.int32(0))   # one histogram per device
        ctx.map(LMOSEM_ORDER_HIST, events, None, args=[hist, *self.dims_args, np.int32(nb)])
        hist.mark_device_modified()              # per-device counts (diverged copies)
        ctx.scan(SUM_I32, hist, cursor, np.int32(0))  # each device scans its own counts
        ctx.map(LMOSEM_ORDER_SCATTER, events, None, args=[cursor, out, *self.dims_args, np.int32(nb)])
        cursor.mark_device_modified()
        out.mark_device_modified()
        return out

    # ---- Listing 4's loop body -------------------------------------------------
    def error_map(self, events: skel.Vector):
        """The error-image Map c += ... over the (already ordered) events."""
        ctx, f, c = self.ctx, self.f, self.c
        src, lanes = self.plan(self.per_device(events))
        ctx.set_block_size(MAP_BLOCK)
        try:
            if lanes == 1:
                ctx.map(src, events, None, args=[f, c, *self.dims_args])
            else:
                ctx.map_lanes(src, events, None, lanes, args=[f, c, *self.dims_args])
        finally:
            ctx.set_block_size(0)

    def subset(self, events: skel.Vector, fused: bool = False):
        """One iteration of Listing 4's loop body.  fused=True runs the tail
        (combine c, update f, redistribute f) as one peer-memory kernel."""
        ctx, f, c = self.ctx, self.f, self.c
        f.set_distribution(skel.COPY)                     # block -> copy: all-gather (no-op after a fused tail)
        c.fill_dist(skel.COPY, np.float32(0))             # fresh zero copy on every device
        ev = self.order_on_device(events) if self.ordered(self.per_device(events)) else events
        self.error_map(ev)
        c.mark_device_modified()                          # dataOnDevicesModified()
        if fused:
            ctx.zip_combine(LMOSEM_UPDATE, f, c, skel.COMBINE_ADD, f)
            return
        f.set_distribution(skel.BLOCK)                    # copy -> block: local slice
        c.set_distribution(skel.BLOCK, skel.COMBINE_ADD)  # copy -> block + add: reduce-scatter
        ctx.zip(LMOSEM_UPDATE, f, c, f)                   # f[j] *= c[j] where c[j] > 0

    def image(self) -> np.ndarray:
        return self.f.download()
