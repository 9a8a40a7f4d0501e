"""GPU parity of list-mode OSEM (§IV-B, Listings 3/4): the
event-parallel Siddon walk Map with scatter-add into the copy-distributed
error image, the copy->block+add combine, and the update Zip.

Bar (north_star): relative L2 error <= 1e-4 of the GPU image against the
oracle (float atomics make the summation order vary), plus closed forms."""
import numpy as np
import pytest

import oracle
import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.lmosem import LMOSEM
from paper_conf_ipps_steuwerkg11_b200.workloads import LMOSEM_ERROR

pytestmark = pytest.mark.gpu


def rel_l2(a, b):
    a = np.asarray(a, np.float64)
    b = np.asarray(b, np.float64)
    return float(np.linalg.norm(a - b) / np.linalg.norm(b))


def ev(*rays):
    e = np.zeros(len(rays), si.EVENT_DTYPE)
    for i, (p1, p2) in enumerate(rays):
        for k, v in zip(("x1", "y1", "z1", "x2", "y2", "z2"), (*p1, *p2)):
            e[k][i] = v
    return e


def error_image(ctx, events, f, dims):
    fv = ctx.vector(f.astype(np.float32))
    c = ctx.vector(n=int(np.prod(dims)), dtype=np.float32)
    ctx.map(LMOSEM_ERROR, ctx.vector(events), None, args=[fv, c, *[np.int32(d) for d in dims]])
    c.mark_device_modified()
    return c.download()


def test_single_event_closed_forms():
    with skel.Context(1) as ctx:
        c = error_image(ctx, ev(((-1, 0.5, 0.5), (5, 3.5, 0.5))), np.ones(16), (4, 4, 1))
        want = np.zeros(16)
        want[[4, 5, 10, 11]] = 0.25
        assert np.allclose(c, want, atol=1e-6)
        c = error_image(ctx, ev(((0, 0, 0), (3, 3, 3))), np.ones(27), (3, 3, 3))
        want = np.zeros(27)
        want[[0, 13, 26]] = 1 / 3
        assert np.allclose(c, want, atol=1e-6)
        # a line that misses the volume contributes nothing
        c = error_image(ctx, ev(((0.5, 0.5, -1), (0.5, 0.5, -5))), np.ones(8), (2, 2, 2))
        assert not c.any()


def test_random_rays_tiny_grid_match_oracle():
    g = np.random.default_rng(1)
    dims = (4, 3, 5)
    n = 400
    e = np.zeros(n, si.EVENT_DTYPE)
    for k in ("x1", "y1", "z1", "x2", "y2", "z2"):
        e[k] = g.uniform(-2, 7, n)
    f = g.uniform(0.5, 2.0, int(np.prod(dims)))
    with skel.Context(1) as ctx:
        c = error_image(ctx, e, f, dims)
    want, _ = oracle.lmosem_error_image(e, f.astype(np.float32).astype(np.float64), dims)
    assert rel_l2(c, want) <= 1e-5


@pytest.mark.parametrize("D", [1, 2, 4, 8])
def test_subset_matches_oracle(D):
    n = 20_000
    events = si.lmosem_events(n, subset=2)
    with skel.Context(D) as ctx:
        rec = LMOSEM(ctx)
        rec.subset(rec.events(events))
        f = rec.image()
    want, c, nv = oracle.lmosem_subset(events, np.ones(150 * 150 * 280))
    assert rel_l2(f, want) <= 1e-4
    # count preservation (Listing 3 identity): sum of updated voxels = #events
    assert abs(float(f[c > 0].astype(np.float64).sum()) - nv) <= 1e-4 * nv


def test_two_subsets_virtual_devices_agree_with_one_device():
    subsets = [si.lmosem_events(10_000, subset=l) for l in range(2)]
    imgs = []
    for D in (1, 4):
        with skel.Context(D) as ctx:
            rec = LMOSEM(ctx)
            for s in subsets:
                rec.subset(rec.events(s))
            imgs.append(rec.image())
    want = oracle.lmosem_reconstruct(subsets)
    assert rel_l2(imgs[0], want) <= 1e-4
    assert rel_l2(imgs[1], want) <= 1e-4
    assert rel_l2(imgs[1], imgs[0]) <= 1e-5


def test_full_size_subset_matches_oracle():
    """Config 4 at its full size: 10^6 events, 150x150x280 voxels."""
    events = si.lmosem_events(1_000_000, subset=0)
    with skel.Context(1) as ctx:
        rec = LMOSEM(ctx)
        rec.subset(rec.events(events))
        f = rec.image()
    want, c, nv = oracle.lmosem_subset(events, np.ones(150 * 150 * 280))
    assert rel_l2(f, want) <= 1e-4
    assert abs(float(f[c > 0].astype(np.float64).sum()) - nv) <= 1e-4 * nv


@pytest.mark.parametrize("n,D", [(1_000_000, 1), (60_000, 4), (20_001, 8)])
def test_device_ordered_events_match_oracle_in_given_order(n, D):
    """order="device": each device's events reordered longest path first on the
    device (counting Map, Scan, scattering Map; workloads/lmosem_order.cu) --
    the oracle's image for the events in their given order (the error image is
    a sum over events, R10(x)), with both Map forms the policy picks."""
    events = si.lmosem_events(n, subset=3)
    with skel.Context(D) as ctx:
        rec = LMOSEM(ctx, order="device")
        rec.subset(rec.events(events))
        f = rec.image()
    want, c, nv = oracle.lmosem_subset(events, np.ones(150 * 150 * 280))
    assert rel_l2(f, want) <= 1e-4
    assert abs(float(f[c > 0].astype(np.float64).sum()) - nv) <= 1e-4 * nv


@pytest.mark.parametrize("D", [1, 3])
def test_device_order_is_a_per_device_permutation_by_bucket(D):
    """The reordered vector holds, on every device, a permutation of that
    device's own events, and their length buckets never increase along it
    (bucket of an event recomputed on the host from the oracle's exact path:
    longer paths first, up to bucket-boundary rounding)."""
    from paper_conf_ipps_steuwerkg11_b200.workloads import LMOSEM_ORDER_BUCKETS
    n = 30_011
    events = si.lmosem_events(n, subset=9)
    with skel.Context(D) as ctx:
        rec = LMOSEM(ctx, order="device")
        ev = rec.events(events)
        out = rec.order_on_device(ev).download()
        parts = [ev.part(k) for k in range(D)]
    rows = lambda a: sorted(map(bytes, a.view(np.uint8).reshape(len(a), -1)))  # noqa: E731
    nb = LMOSEM_ORDER_BUCKETS
    for lo, hi in parts:
        assert rows(out[lo:hi]) == rows(events[lo:hi])
        seg = out[lo:hi]
        nvox = np.array([len(oracle.compute_path((e["x1"], e["y1"], e["z1"]), (e["x2"], e["y2"], e["z2"]))[0])
                         for e in seg[:: max(1, len(seg) // 2000)]])
        # the oracle's voxel count per path decreases along the order
        from scipy.stats import spearmanr
        r = spearmanr(np.arange(len(nvox)), nvox).statistic
        assert r < -0.95, r
    assert nb >= 16


@pytest.mark.parametrize("lanes", [1, 2, 4, 8, 32])
def test_lanes_map_error_image_matches_oracle(lanes):
    """The error image on a lanes Map (skel_map_lanes: `lanes` threads per
    event, each walking an alpha piece of the line of response, the partial
    forward projections summed over the group): the oracle's image (relL2 1e-4
    bar; here 1e-5 on a random tiny grid with ties and at the paper's volume)."""
    from paper_conf_ipps_steuwerkg11_b200.workloads import LMOSEM_LANES
    g = np.random.default_rng(3)
    dims = (4, 3, 5)
    n = 600
    e = np.zeros(n, si.EVENT_DTYPE)
    for k in ("x1", "y1", "z1", "x2", "y2", "z2"):
        e[k] = g.integers(-8, 28, n) / 4.0
    f = g.uniform(0.5, 2.0, int(np.prod(dims))).astype(np.float32)
    events = si.lmosem_events(50_003, subset=7)
    with skel.Context(1) as ctx:
        for evs, ff, dd in ((e, f, dims), (events, np.ones(150 * 150 * 280, np.float32), (150, 150, 280))):
            fv = ctx.vector(ff)
            c = ctx.vector(n=int(np.prod(dd)), dtype=np.float32)
            ctx.map_lanes(LMOSEM_LANES, ctx.vector(evs), None, lanes, args=[fv, c, *[np.int32(d) for d in dd]])
            c.mark_device_modified()
            got = c.download()
            want, _ = oracle.lmosem_error_image(evs, ff.astype(np.float64), dd)
            assert np.array_equal(got > 0, want > 0)
            assert rel_l2(got, want) <= 1e-5


def test_lanes_map_generic_group_sum():
    """skel_map_lanes semantics on a plain function: lane l of element x
    contributes x * (l + 1); the group sum is x * lanes (lanes + 1) / 2 in every
    lane, lane 0's result is stored (eq. (1) with a cooperative element)."""
    src = """
    float tri(float x, int lane, int lanes) {
        return skel_group_sum(x * (float)(lane + 1), lanes);
    }"""
    x = np.arange(1, 10_001, dtype=np.float32)
    with skel.Context(1) as ctx:
        vx = ctx.vector(x)
        out = ctx.vector(n=x.size, dtype=np.float32)
        for lanes in (1, 2, 4, 8, 16, 32):
            ctx.map_lanes(src, vx, out, lanes)
            assert np.array_equal(out.download(), x * np.float32(lanes * (lanes + 1) // 2))
        with pytest.raises(skel.SkelError) as e:
            ctx.map_lanes(src, vx, out, 3)
        assert e.value.name == "SKEL_ERR_ARG"
