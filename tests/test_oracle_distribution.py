"""Pins for the oracle's distribution model (§III-D, Listing 4)."""
import numpy as np
import pytest

from oracle import distribution as dist


@pytest.mark.parametrize("n,D", [(0, 1), (1, 4), (7, 2), (10, 4), (6_300_000, 8), (5, 8)])
def test_parts_cover_disjointly(n, D):
    ranges = [dist.part_range(n, D, k) for k in range(D)]
    assert ranges[0][0] == 0 and ranges[-1][1] == n
    for (a, b), (c, d) in zip(ranges, ranges[1:]):
        assert b == c and a <= b
    if n % D == 0:
        assert all(b - a == n // D for a, b in ranges)


def test_paper_image_parts_are_z_slabs():
    # 150*150*280 voxels on 8 devices: 787,500 = 150*150*35 per part
    assert dist.part_range(150 * 150 * 280, 8, 1) == (787_500, 1_575_000)


@pytest.mark.parametrize("D", [1, 2, 3, 4, 8])
def test_round_trips_identity(D):
    x = np.arange(37, dtype=np.int32)
    for a in (dist.SINGLE, dist.BLOCK, dist.COPY):
        for b in (dist.SINGLE, dist.BLOCK, dist.COPY):
            p = dist.distribute(x, a, D)
            q = dist.redistribute(dist.redistribute(p, a, b), b, a)
            assert np.array_equal(dist.gather(q, a), x)


@pytest.mark.parametrize("D", [1, 2, 4, 8])
def test_copy_to_block_add_of_equal_copies(D):
    x = np.arange(29, dtype=np.float64)
    p = dist.redistribute(dist.distribute(x, dist.COPY, D), dist.COPY, dist.BLOCK, "add")
    assert np.array_equal(np.concatenate(p), D * x)


def test_copy_to_block_add_of_distinct_copies():
    copies = [np.full(6, float(d + 1)) for d in range(3)]  # 1, 2, 3
    p = dist.redistribute(copies, dist.COPY, dist.BLOCK, "add")
    assert [a.tolist() for a in p] == [[6.0, 6.0], [6.0, 6.0], [6.0, 6.0]]


def test_copy_to_block_without_combine_is_local_slice():
    copies = [np.full(4, float(d)) for d in range(2)]
    p = dist.redistribute(copies, dist.COPY, dist.BLOCK)
    assert [a.tolist() for a in p] == [[0.0, 0.0], [1.0, 1.0]]


def test_combine_requires_copy_source():
    with pytest.raises(ValueError):
        dist.redistribute(dist.distribute(np.ones(4), dist.BLOCK, 2), dist.BLOCK, dist.COPY, "add")
