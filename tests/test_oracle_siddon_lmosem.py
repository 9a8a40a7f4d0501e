"""Pins for the oracle's compute_path (Siddon) and LM OSEM (Listing 3).

compute_path is checked against a brute-force per-voxel slab clip in exact
rational arithmetic (a different algorithm from the oracle's merged-alpha
walk), against hand-worked rays and against invariants.  LM OSEM is checked
against single-event closed forms worked by hand and the count-preservation
identity sum_j f_j c_j = #events (exact in real arithmetic).
"""
import math
from fractions import Fraction

import numpy as np
import pytest

import oracle
from skel_inputs import EVENT_DTYPE, NX, NY, NZ, lmosem_events


def brute_path(p1, p2, dims):
    """{coord: length} by clipping the segment against every voxel box exactly."""
    P1 = [Fraction(float(v)) for v in p1]
    P2 = [Fraction(float(v)) for v in p2]
    d = [b - a for a, b in zip(P1, P2)]
    L = math.sqrt(sum(float(v) ** 2 for v in d))
    nx, ny, nz = dims
    out = {}
    for k in range(nz):
        for j in range(ny):
            for i in range(nx):
                t0, t1 = Fraction(0), Fraction(1)
                ok = True
                for a, lo in enumerate((i, j, k)):
                    hi = lo + 1
                    if d[a] == 0:
                        if not (lo <= P1[a] < hi):
                            ok = False
                            break
                        continue
                    ta, tb = (lo - P1[a]) / d[a], (hi - P1[a]) / d[a]
                    if ta > tb:
                        ta, tb = tb, ta
                    t0, t1 = max(t0, ta), min(t1, tb)
                if ok and t1 > t0:
                    out[i + nx * (j + ny * k)] = float(t1 - t0) * L
    return out


def as_dict(coords, lens):
    assert len(set(coords.tolist())) == len(coords), "a voxel appears twice on one line"
    return dict(zip(coords.tolist(), lens.tolist()))


def assert_paths_equal(got, want):
    assert set(got) == set(want)
    for k in want:
        assert got[k] == pytest.approx(want[k], rel=1e-12, abs=1e-12)


# ---- hand-worked rays -----------------------------------
def test_ray_through_corners():
    # (-1,1/2,1/2) -> (5,7/2,1/2) in 4x4x1 passes the corners (0,1) and (2,2)
    c, l = oracle.compute_path((-1, 0.5, 0.5), (5, 3.5, 0.5), (4, 4, 1))
    assert c.tolist() == [4, 5, 10, 11]
    assert np.allclose(l, math.sqrt(1.25), rtol=0, atol=1e-14)


def test_axis_parallel_ray():
    c, l = oracle.compute_path((-2, 0.5, 0.5), (6, 0.5, 0.5), (4, 4, 1))
    assert c.tolist() == [0, 1, 2, 3] and np.allclose(l, 1.0)


def test_body_diagonal():
    c, l = oracle.compute_path((0, 0, 0), (3, 3, 3), (3, 3, 3))
    assert c.tolist() == [0, 13, 26] and np.allclose(l, math.sqrt(3))


def test_miss_and_half_open_planes():
    assert oracle.compute_path((0.5, 0.5, -1), (0.5, 0.5, -5), (2, 2, 2))[0].size == 0
    # a line in the plane x = 2 belongs to voxels with i = 2 (lo <= p < hi)
    c, _ = oracle.compute_path((2, -1, 0.5), (2, 5, 0.5), (4, 4, 1))
    assert c.tolist() == [2, 6, 10, 14]
    # ... and the plane x = nx is outside
    assert oracle.compute_path((4, -1, 0.5), (4, 5, 0.5), (4, 4, 1))[0].size == 0


def test_segment_semantics_endpoint_inside():
    c, l = oracle.compute_path((0.5, 0.5, 0.5), (2.5, 0.5, 0.5), (4, 1, 1))
    assert c.tolist() == [0, 1, 2] and np.allclose(l, [0.5, 1.0, 0.5])


# ---- brute force on tiny grids ---------------------------------------------
@pytest.mark.parametrize("seed", range(6))
def test_brute_force_random_rays(seed):
    g = np.random.default_rng(seed)
    dims = (4, 3, 5)
    for t in range(40):
        if t % 2:   # quarter-grid endpoints: many exact plane/edge/corner ties
            p1 = g.integers(-8, 28, 3) / 4.0
            p2 = g.integers(-8, 28, 3) / 4.0
        else:
            p1 = g.uniform(-2, 7, 3)
            p2 = g.uniform(-2, 7, 3)
        got = as_dict(*oracle.compute_path(p1, p2, dims))
        want = brute_path(p1, p2, dims)
        assert_paths_equal(got, want)


# ---- invariants on the paper-sized grid -------------------------------------
def test_invariants_full_grid():
    ev = lmosem_events(300, subset=3)
    for e in ev:
        p1 = np.array([e["x1"], e["y1"], e["z1"]], np.float64)
        p2 = np.array([e["x2"], e["y2"], e["z2"]], np.float64)
        c, l = oracle.compute_path(p1, p2, (NX, NY, NZ))
        assert len(c) <= NX + NY + NZ - 2
        assert np.all(l > 0) and np.all((c >= 0) & (c < NX * NY * NZ))
        # sum of lengths = length of the chord clipped to the box (slab clip, closed form)
        d = p2 - p1
        t0, t1 = 0.0, 1.0
        for a, n in enumerate((NX, NY, NZ)):
            ta, tb = sorted(((0 - p1[a]) / d[a], (n - p1[a]) / d[a]))
            t0, t1 = max(t0, ta), min(t1, tb)
        chord = max(0.0, t1 - t0) * np.linalg.norm(d)
        assert l.sum() == pytest.approx(chord, rel=1e-12, abs=1e-9)
        # reversing the ray gives the same multiset
        c2, l2 = oracle.compute_path(p2, p1, (NX, NY, NZ))
        assert_paths_equal(as_dict(c2, l2), as_dict(c, l))


# ---- LM OSEM, Listing 3 -----------------------------------------------------
def _ev(p1, p2):
    e = np.zeros(1, EVENT_DTYPE)
    for k, v in zip(("x1", "y1", "z1", "x2", "y2", "z2"), (*p1, *p2)):
        e[k] = v
    return e


def test_single_event_uniform_image():
    # f = 1: fp = sum(len) = 4 sqrt(1.25); c_v = len_v / fp = 1/4 on the path
    dims = (4, 4, 1)
    f = np.ones(16)
    fn, c, nv = oracle.lmosem_subset(_ev((-1, 0.5, 0.5), (5, 3.5, 0.5)), f, dims)
    assert nv == 1
    want = np.zeros(16)
    want[[4, 5, 10, 11]] = 0.25
    assert np.allclose(c, want, atol=1e-15)
    assert np.allclose(fn, np.where(want > 0, 0.25, 1.0), atol=1e-15)


def test_single_event_nonuniform_image():
    # f = 2 on voxel 4: fp = 5 sqrt(1.25); c = 1/5 on the path; f_new[4] = 0.4, others 0.2
    dims = (4, 4, 1)
    f = np.ones(16)
    f[4] = 2.0
    fn, c, _ = oracle.lmosem_subset(_ev((-1, 0.5, 0.5), (5, 3.5, 0.5)), f, dims)
    assert np.allclose(c[[4, 5, 10, 11]], 0.2) and c.sum() == pytest.approx(0.8)
    assert fn[4] == pytest.approx(0.4) and fn[5] == pytest.approx(0.2) and fn[0] == 1.0


def test_diagonal_event_thirds_and_missing_event_skipped():
    dims = (3, 3, 3)
    ev = np.concatenate([_ev((0, 0, 0), (3, 3, 3)), _ev((0.5, 0.5, -1), (0.5, 0.5, -5))])
    c, nv = oracle.lmosem_error_image(ev, np.ones(27), dims)
    assert nv == 1
    assert np.allclose(c[[0, 13, 26]], 1 / 3) and c.sum() == pytest.approx(1.0)


def test_update_only_where_c_positive():
    f = np.array([1.0, 2.0, 3.0])
    assert oracle.lmosem_update(f, np.array([0.5, 0.0, -1.0])).tolist() == [0.5, 2.0, 3.0]


def test_count_preservation_full_grid():
    """sum_j f_j c_j = sum_e sum_m f[v_m] len_m / fp_e = N_valid, and after the
    update sum_{c_j>0} f_j^new equals it too (exact in real arithmetic)."""
    ev = lmosem_events(3000, subset=1)
    g = np.random.default_rng(0)
    f = g.uniform(0.5, 2.0, NX * NY * NZ)
    c, nv = oracle.lmosem_error_image(ev, f)
    assert nv == 3000  # every generated line crosses the phantom volume
    assert float(np.dot(f, c)) == pytest.approx(nv, rel=1e-10)
    fn = oracle.lmosem_update(f, c)
    assert float(fn[c > 0].sum()) == pytest.approx(nv, rel=1e-10)
    assert np.all(fn > 0)


def test_two_subset_reconstruction_positive_and_preserving():
    subsets = [lmosem_events(1000, subset=l) for l in range(2)]
    f = oracle.lmosem_reconstruct(subsets)
    assert np.all(f > 0)
    # after the last subset, the voxels it touched carry exactly its event count
    f1 = oracle.lmosem_reconstruct(subsets[:1])
    c, nv = oracle.lmosem_error_image(subsets[1], f1)
    assert float(f[c > 0].sum()) == pytest.approx(nv, rel=1e-10)


def test_events_on_detector_cylinder():
    ev = lmosem_events(2000, subset=0)
    for a, b in (("x1", "y1"), ("x2", "y2")):
        r = np.hypot(ev[a].astype(np.float64) - 75, ev[b].astype(np.float64) - 75)
        assert np.allclose(r, 110.0, atol=1e-4)
