"""Pure model of SkelCL vector distributions -- TEST INFRASTRUCTURE ONLY.

PAPER.md §III-D: a Vector is either "completely copied to every
device" (copy) or "evenly divided into one part per device" (block); a
redistribution changes the distribution and moves the data automatically.
Listing 4 adds copy -> block with an element-wise combine of the
per-device copies ("reduce (element-wise add) all copies of error image").
`single` (the whole vector on device 0) comes from the task's north star
(reading R6).

A distributed vector is modelled as a list of D per-device numpy arrays (None
where a device holds nothing).  Every transition is written out directly from
its definition; there is no notion of collectives here.
"""
from __future__ import annotations

import numpy as np

SINGLE, BLOCK, COPY = "single", "block", "copy"


def part_range(n: int, D: int, k: int) -> tuple[int, int]:
    """Part k of a block-distributed vector of n elements on D devices.

    "evenly divided into one part per device"; n mod D != 0 is
    not addressed by the paper -> parts of ceil(n/D), the last ones shorter
    (reading R6(ii)).
    """
    s = -(-n // D) if D > 0 else 0
    lo = min(n, k * s)
    hi = min(n, (k + 1) * s)
    return lo, hi


def distribute(x: np.ndarray, dist: str, D: int) -> list:
    """Place a host vector x on D devices under `dist`."""
    if dist == SINGLE:
        return [x.copy()] + [None] * (D - 1)
    if dist == COPY:
        return [x.copy() for _ in range(D)]
    if dist == BLOCK:
        return [x[slice(*part_range(x.size, D, k))].copy() for k in range(D)]
    raise ValueError(dist)


def gather(parts: list, dist: str) -> np.ndarray:
    """The vector's value as the host sees it after a download.

    copy: device 0's copy (reading R6: a diverged copy is read from device 0).
    """
    if dist in (SINGLE, COPY):
        return parts[0].copy()
    return np.concatenate(parts)


def redistribute(parts: list, src: str, dst: str, combine: str | None = None) -> list:
    """Change the distribution of a vector held as `parts` from src to dst.

    combine = "add" merges the D copies element-wise (Listing 4)
    and is only meaningful from `copy`; a callable f(acc, x) is a user-defined
    element-wise combine, folded over the copies in device order.
    """
    D = len(parts)
    if combine is not None and combine != "add" and not callable(combine):
        raise ValueError(combine)
    if combine is not None and src != COPY:
        raise ValueError("a combine merges per-device copies: source must be copy")
    if src == COPY and combine is not None:
        # element-wise, folded over the copies in device order (a callable is a
        # user combine f(acc, x) applied to whole arrays, NEXT-2)
        f = (lambda a, b: a + b) if combine == "add" else combine
        total = parts[0].copy()
        for d in range(1, D):
            total = f(total, parts[d])
        return distribute(total, dst, D)
    if src == COPY and dst == BLOCK:
        # each device keeps its own slice of its own copy (no data exchange)
        n = parts[0].size
        return [parts[k][slice(*part_range(n, D, k))].copy() for k in range(D)]
    if src == COPY and dst == SINGLE:
        return [parts[0].copy()] + [None] * (D - 1)
    return distribute(gather(parts, src), dst, D)
