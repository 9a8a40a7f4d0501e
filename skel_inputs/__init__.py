"""Seeded synthetic input generators shared by the oracle and the CUDA path.

This module holds NONE of the method's arithmetic (no Map/Zip/Reduce/Scan,
no escape-time iteration, no ray walk, no OSEM update).  It only builds the
input vectors the workloads consume, with the shapes and value distributions
stated in DESIGN.md §3 ("input recipe"):

* skeleton sweep vectors: float32 U[0,1) and int32
  data drawn from PCG64 with seed 20110516 + k;
* Mandelbrot pixel positions ("A Vector of
  complex numbers, each of which is represented by a pixel ... is passed to
  the Map skeleton"), on the window of DESIGN.md reading R5;
* list-mode PET events (~10^7 events, 10
  subsets, 150x150x280 image) drawn from a synthetic phantom (R9).

Both `oracle/` and the product tests/bench import from here; neither side
imports the other.
"""
from __future__ import annotations

import numpy as np

SEED_BASE = 20110516

# Vector<{float re, im}> element of the Mandelbrot Map (8 bytes, AoS).
POS_DTYPE = np.dtype([("re", np.float32), ("im", np.float32)])
# Vector<{Pos, Pos}>: two neighbouring pixels per element (the same bytes as a
# Vector<Pos> of twice the length; workloads/mandelbrot_pairs.cu)
POS2_DTYPE = np.dtype([("re0", np.float32), ("im0", np.float32), ("re1", np.float32), ("im1", np.float32)])
CNT2_DTYPE = np.dtype([("n0", np.int32), ("n1", np.int32)])
# Vector<Event> element of LM OSEM: {float x1,y1,z1,x2,y2,z2} (24 bytes, AoS),
# DESIGN.md reading R8 (PAPER.md P:L520 leaves the fields unspecified).
EVENT_DTYPE = np.dtype([("x1", np.float32), ("y1", np.float32), ("z1", np.float32),
                        ("x2", np.float32), ("y2", np.float32), ("z2", np.float32)])

# PET volume of PAPER.md P:L604 (150 x 150 x 280 voxels), unit voxels.
NX, NY, NZ = 150, 150, 280


def rng(seed: int) -> np.random.Generator:
    return np.random.Generator(np.random.PCG64(seed))


# --------------------------------------------------------------------------
# skeleton sweep data
# --------------------------------------------------------------------------
def uniform_f32(n: int, seed: int) -> np.ndarray:
    """float32 uniform on [0, 1)."""
    return rng(seed).random(n, dtype=np.float32)


def uniform_signed_f32(n: int, seed: int) -> np.ndarray:
    """float32 uniform on [-1, 1): signed Reduce/Scan data (partial sums cancel)."""
    return (rng(seed).random(n, dtype=np.float32) * np.float32(2.0) - np.float32(1.0)).astype(np.float32)


def cancellation_f32(n: int, seed: int) -> np.ndarray:
    """float32 data with catastrophic cancellation: blocks of four
    [s*2^24, u, -s*2^24, u'] (s = +-1 at random, u, u' ~ U[0,1)), truncated to n.
    A float32 left fold loses the small terms next to 2^24; the big ones cancel."""
    g = rng(seed)
    k = (n + 3) // 4
    s = np.where(g.random(k) < 0.5, -1.0, 1.0).astype(np.float32) * np.float32(2.0 ** 24)
    u = g.random((k, 2), dtype=np.float32)
    out = np.stack([s, u[:, 0], -s, u[:, 1]], axis=1).reshape(-1)
    return np.ascontiguousarray(out[:n], dtype=np.float32)


def uniform_int01(n: int, seed: int) -> np.ndarray:
    """int32 uniform on {0, 1}: Reduce/Scan data whose prefix sums never overflow."""
    return rng(seed).integers(0, 2, size=n, dtype=np.int32)


def uniform_i32(n: int, seed: int, lo: int = -(1 << 20), hi: int = (1 << 20)) -> np.ndarray:
    """int32 uniform on [lo, hi): Map/Zip data (saxpy with a=3 cannot overflow)."""
    return rng(seed).integers(lo, hi, size=n, dtype=np.int32)


def uniform_u32(n: int, seed: int) -> np.ndarray:
    """uint32 over the full range: wrap-around (mod 2^32) tests."""
    return rng(seed).integers(0, 1 << 32, size=n, dtype=np.uint64).astype(np.uint32)


# --------------------------------------------------------------------------
# Mandelbrot positions (reading R5)
# --------------------------------------------------------------------------
def mandelbrot_positions(width: int, height: int) -> np.ndarray:
    """Row-major pixel grid, py outer: c = (-2.5 + px*4/W, -1.5 + py*3/H).

    For W in {1024, 4096} and H = 3W/4 the steps 4/W and 3/H are powers of
    two, so every coordinate is an exact float32 (no rounding in this input).
    """
    px = np.arange(width, dtype=np.float64)
    py = np.arange(height, dtype=np.float64)
    re = -2.5 + px * (4.0 / width)
    im = -1.5 + py * (3.0 / height)
    out = np.empty((height, width), dtype=POS_DTYPE)
    out["re"] = re[None, :].astype(np.float32)
    out["im"] = im[:, None].astype(np.float32)
    return out.reshape(-1)


# --------------------------------------------------------------------------
# LM OSEM events (reading R9): phantom + detector cylinder
# --------------------------------------------------------------------------
CYL_CENTER = (75.0, 75.0)
CYL_RADIUS = 60.0
CYL_Z = (15.0, 265.0)
HOT_SPHERES = [((75.0, 45.0, 140.0), 10.0), ((105.0, 75.0, 100.0), 10.0),
               ((60.0, 95.0, 200.0), 10.0)]
HOT_ACTIVITY = 4.0
COLD_SPHERE = ((50.0, 60.0, 70.0), 12.0)
DETECTOR_RADIUS = 110.0  # encloses the volume corners (distance 106.07)
COS_THETA_MAX = 0.3


def phantom_activity(p: np.ndarray) -> np.ndarray:
    """Emission density of the synthetic phantom at points p (k x 3)."""
    x, y, z = p[:, 0], p[:, 1], p[:, 2]
    inside = ((x - CYL_CENTER[0]) ** 2 + (y - CYL_CENTER[1]) ** 2 <= CYL_RADIUS ** 2) & \
             (z >= CYL_Z[0]) & (z < CYL_Z[1])
    act = np.where(inside, 1.0, 0.0)
    for (cx, cy, cz), r in HOT_SPHERES:
        hot = (x - cx) ** 2 + (y - cy) ** 2 + (z - cz) ** 2 <= r * r
        act = np.where(hot & inside, HOT_ACTIVITY, act)
    (cx, cy, cz), r = COLD_SPHERE
    cold = (x - cx) ** 2 + (y - cy) ** 2 + (z - cz) ** 2 <= r * r
    return np.where(cold, 0.0, act)


def lmosem_events(n: int, subset: int = 0, seed_base: int = SEED_BASE) -> np.ndarray:
    """n list-mode events (lines of response) of subset `subset`.

    Emission points are rejection-sampled from the phantom; each event's
    direction has phi ~ U[0, 2pi) and cos(theta) ~ U[-0.3, 0.3] (theta from
    the scanner axis z); the two endpoints are the intersections of that line
    with the detector cylinder of radius 110 around the volume axis.
    Coordinates are voxel units; the volume is [0,150)x[0,150)x[0,280).
    """
    g = rng(seed_base + subset)
    pts = np.empty((0, 3))
    x0, y0 = CYL_CENTER
    while len(pts) < n:
        k = max(2 * (n - len(pts)), 1024)
        cand = np.stack([g.uniform(x0 - CYL_RADIUS, x0 + CYL_RADIUS, k),
                         g.uniform(y0 - CYL_RADIUS, y0 + CYL_RADIUS, k),
                         g.uniform(CYL_Z[0], CYL_Z[1], k)], axis=1)
        keep = g.uniform(0.0, HOT_ACTIVITY, k) < phantom_activity(cand)
        pts = np.concatenate([pts, cand[keep]])
    pts = pts[:n]
    phi = g.uniform(0.0, 2.0 * np.pi, n)
    ct = g.uniform(-COS_THETA_MAX, COS_THETA_MAX, n)
    st = np.sqrt(1.0 - ct * ct)
    u = np.stack([st * np.cos(phi), st * np.sin(phi), ct], axis=1)
    qx, qy = pts[:, 0] - x0, pts[:, 1] - y0
    a = u[:, 0] ** 2 + u[:, 1] ** 2
    b = qx * u[:, 0] + qy * u[:, 1]
    c = qx * qx + qy * qy - DETECTOR_RADIUS ** 2
    disc = np.sqrt(b * b - a * c)
    t1 = (-b - disc) / a
    t2 = (-b + disc) / a
    p1 = pts + t1[:, None] * u
    p2 = pts + t2[:, None] * u
    ev = np.empty(n, dtype=EVENT_DTYPE)
    for j, name in enumerate(("x1", "y1", "z1")):
        ev[name] = p1[:, j].astype(np.float32)
    for j, name in enumerate(("x2", "y2", "z2")):
        ev[name] = p2[:, j].astype(np.float32)
    return ev


def lmosem_subsets(n_events: int, n_subsets: int = 10) -> list[np.ndarray]:
    """The paper's data set split into equally sized subsets."""
    per = n_events // n_subsets
    return [lmosem_events(per, subset=l) for l in range(n_subsets)]
