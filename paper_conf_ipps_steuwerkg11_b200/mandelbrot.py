"""Mandelbrot images on the skeletons (§IV-A, eq. (5)) with cyclic
rows.

The paper block-distributes the image's rows (4096x3072 on up to
4 GPUs), which leaves the device holding the middle rows with most
of the work (3.1x the mean at 8 devices).  `cyclic_image` gives device k the
rows k, k+D, k+2D, ... instead -- with no new distribution type: an index Map
computes the image in a permuted row order into a block-distributed vector
(workloads/mandelbrot_cyclic.cu), the parts are gathered on device 0
(block -> single), and a second index Map restores row-major order
(workloads/mandelbrot_unpermute.cu).  Counts are bit-identical to eq. (5) as
written (two pixels per element, packed arithmetic: mandelbrot_pairs.cu).
"""
from __future__ import annotations

import numpy as np

from . import skel
from .workloads import MANDELBROT_CYCLIC, MANDELBROT_UNPERMUTE

CNT2 = np.dtype([("n0", np.int32), ("n1", np.int32)])


class CyclicMandelbrot:
    """Reusable buffers for `image` at one size (W must be even)."""

    def __init__(self, ctx: skel.Context, width: int, height: int):
        if width % 2:
            raise ValueError("cyclic rows process two pixels per element: the width must be even")
        self.ctx, self.W, self.H = ctx, int(width), int(height)
        D = ctx.D
        self.R = -(-self.H // D)                     # row slots per device
        self.n_perm = D * self.R * self.W // 2       # pixel pairs of the permuted image (padded)
        self.perm = ctx.vector(n=self.n_perm, dtype=CNT2)
        self.out = ctx.vector(n=self.H * self.W // 2, dtype=CNT2)
        self.out.fill_dist(skel.SINGLE, np.zeros(1, CNT2)[0])

    def compute(self, cap: int):
        """The permuted image, block-distributed: device k computes rows k, k+D, ..."""
        D = self.ctx.D
        self.perm.fill_dist(skel.BLOCK if D > 1 else skel.SINGLE, np.zeros(1, CNT2)[0])
        self.ctx.map_index(MANDELBROT_CYCLIC, self.n_perm, self.perm,
                           args=[np.int32(self.W), np.int32(self.H), np.int32(cap), np.int32(D)])

    def image(self, cap: int) -> skel.Vector:
        """Row-major counts (pairs of int32) on device 0 (single distribution)."""
        self.compute(cap)
        self.perm.set_distribution(skel.SINGLE)     # block -> single: gather on device 0
        self.ctx.map_index(MANDELBROT_UNPERMUTE, self.H * self.W // 2, self.out,
                           args=[self.perm, np.int32(self.W), np.int32(self.H), np.int32(self.ctx.D)])
        return self.out

    def counts(self, cap: int) -> np.ndarray:
        return self.image(cap).download().view(np.int32)
