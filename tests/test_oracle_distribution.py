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


@pytest.mark.parametrize("D", [2, 3, 5])
def test_user_combine_folds_in_device_order(D):
    """NEXT-2 user combine: element-wise fold over the copies in device order.
    Pinned by 2x2 integer matrix products (associative, not commutative):
    folding copy d = [[1, d+1], [0, 1]] gives [[1, D(D+1)/2], [0, 1]], and
    reversing the order of non-commuting factors changes the result."""
    n = 4
    copies = []
    for d in range(D):
        m = np.zeros((n, 2, 2), dtype=np.int64)
        m[:, 0, 0] = m[:, 1, 1] = 1
        m[:, 0, 1] = d + 1
        copies.append(m)
    matmul = lambda a, b: np.einsum("nij,njk->nik", a, b)
    out = dist.gather(dist.redistribute(copies, dist.COPY, dist.BLOCK, matmul), dist.BLOCK)
    assert (out[:, 0, 1] == D * (D + 1) // 2).all() and (out[:, 0, 0] == 1).all() and (out[:, 1, 0] == 0).all()
    # a non-commuting case: upper- then lower-triangular differs from the reverse
    u = np.array([[[1, 1], [0, 1]]] * n)
    low = np.array([[[1, 0], [1, 1]]] * n)
    fwd = dist.gather(dist.redistribute([u, low], dist.COPY, dist.SINGLE, matmul), dist.SINGLE)
    rev = dist.gather(dist.redistribute([low, u], dist.COPY, dist.SINGLE, matmul), dist.SINGLE)
    assert fwd[0].tolist() == [[2, 1], [1, 1]] and rev[0].tolist() == [[1, 1], [1, 2]]


def test_user_add_equals_builtin_add():
    parts = [np.arange(10, dtype=np.int32) * (d + 1) for d in range(3)]
    a = dist.redistribute(parts, dist.COPY, dist.COPY, "add")
    b = dist.redistribute(parts, dist.COPY, dist.COPY, lambda x, y: x + y)
    assert all(np.array_equal(p, q) for p, q in zip(a, b))
