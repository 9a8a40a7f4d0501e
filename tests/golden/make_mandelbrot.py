"""Regenerate tests/golden/mandelbrot.json -- the whole-image Mandelbrot pins.

An implementation of eq. (5) written directly in numpy
float32, independent of oracle/ (it imports neither oracle/ nor the product):
z_0 = 0, z_{i+1} = z_i^2 + c; the count is the number of updates made before
x*x + y*y > 4 or the cap is reached (reading R4).  The window is
reading R5: c = (-2.5 + px*4/W, -1.5 + py*3/H), row-major, py outer; for
W in {1024, 4096} every c is an exact float32.  numpy evaluates each
elementwise float32 operation separately with round-to-nearest-even (no FMA
contraction), in exactly the operation order of the oracle's loop:
xt = (x*x - y*y) + cx; y = (2*x)*y + cy; x = xt.

    python tests/golden/make_mandelbrot.py          # check against the stored pins
    python tests/golden/make_mandelbrot.py --write  # rewrite mandelbrot.json

CRC32 = zlib.crc32 of the int32 little-endian row-major counts.
"""
from __future__ import annotations

import json
import sys
import zlib
from pathlib import Path

import numpy as np

HERE = Path(__file__).resolve().parent
CASES = [(1024, 768, 256), (4096, 3072, 256), (1024, 768, 4096)]


def counts(width: int, height: int, cap: int, rows_per_block: int = 256) -> np.ndarray:
    f = np.float32
    px = np.arange(width, dtype=np.float64)
    re_row = (-2.5 + px * (4.0 / width)).astype(f)
    out = np.empty((height, width), np.int32)
    for r0 in range(0, height, rows_per_block):
        r1 = min(height, r0 + rows_per_block)
        py = np.arange(r0, r1, dtype=np.float64)
        cy = np.broadcast_to((-1.5 + py * (3.0 / height)).astype(f)[:, None], (r1 - r0, width)).copy()
        cx = np.broadcast_to(re_row[None, :], (r1 - r0, width)).copy()
        x = np.zeros_like(cx)
        y = np.zeros_like(cx)
        n = np.zeros(cx.shape, np.int32)
        live = np.ones(cx.shape, bool)
        two, four = f(2.0), f(4.0)
        for _ in range(cap):
            # loop condition of the current iterate: n < cap and |z|^2 <= 4
            live &= (x * x + y * y) <= four
            if not live.any():
                break
            xt = (x * x - y * y) + cx
            yn = (two * x) * y + cy
            x = np.where(live, xt, x)
            y = np.where(live, yn, y)
            n += live
        out[r0:r1] = n
    return out.reshape(-1)


def pins(width: int, height: int, cap: int) -> dict:
    c = counts(width, height, cap)
    d = {"width": width, "height": height, "cap": cap, "sum_iter": int(c.sum(dtype=np.int64))}
    if cap == 256:
        d["at_cap"] = int((c == cap).sum())
    d["crc32"] = f"0x{zlib.crc32(c.astype('<i4').tobytes()) & 0xffffffff:08x}"
    return d


def main() -> int:
    path = HERE / "mandelbrot.json"
    stored = json.loads(path.read_text())
    fresh = [pins(*c) for c in CASES]
    if "--write" in sys.argv:
        stored["cases"] = fresh
        path.write_text(json.dumps(stored, indent=2) + "\n")
        print("wrote", path)
        return 0
    ok = True
    for want, got in zip(stored["cases"], fresh):
        same = all(want[k] == got[k] for k in want)
        ok &= same
        print(("OK  " if same else "DIFF"), got)
    return 0 if ok else 1


if __name__ == "__main__":
    sys.exit(main())
