"""Pins for the oracle's Mandelbrot escape-time count (eq. (5)).

Readings (R4/R5): z_0 = 0, z_{i+1} = z_i^2 + c; the count is the
number of updates made while |z|^2 <= 4, capped at `cap`; float32, no FMA.
"""
import json
import os
import zlib
from decimal import Decimal, getcontext

import numpy as np
import pytest

import oracle
from skel_inputs import POS_DTYPE, mandelbrot_positions


def _pts(cs):
    p = np.zeros(len(cs), POS_DTYPE)
    p["re"] = [c.real for c in cs]
    p["im"] = [c.imag for c in cs]
    return p


# Closed forms, worked by hand (orbits in exact arithmetic):
#   c=1: 0 -> 1 -> 2 -> 5: |z_2|^2 = 4 is not > 4, so the third update happens -> 3
#   c=2: 0 -> 2 -> 6 -> 2
#   c=-1.5+1.5i: |z_1|^2 = 4.5 > 4 -> 1
#   c=0, -1 (0,-1,0,-1 ...), -2 (0,-2,2,2,...: |z|^2 = 4 exactly, the '<=' tie),
#   i (0, i, -1+i, -i, -1+i, ...), 0.25 (increases to the parabolic point 1/2): members -> cap
CLOSED = [(1 + 0j, 3), (2 + 0j, 2), (-1.5 + 1.5j, 1), (0j, 256), (-1 + 0j, 256),
          (-2 + 0j, 256), (1j, 256), (0.25 + 0j, 256), (3 + 0j, 1), (-3 + 0j, 1)]


def test_closed_form_points():
    cs = [c for c, _ in CLOSED]
    got = oracle.mandelbrot(_pts(cs), 256)
    assert got.tolist() == [k for _, k in CLOSED]


def test_cap_is_respected():
    got = oracle.mandelbrot(_pts([0j, 1 + 0j]), 7)
    assert got.tolist() == [7, 3]
    assert oracle.mandelbrot(_pts([0j]), 0).tolist() == [0]


def _decimal_count(cr, ci, cap, digits=80):
    """High-precision escape count and the smallest |(|z|^2 - 4)| margin seen."""
    getcontext().prec = digits
    cr, ci = Decimal(float(cr)), Decimal(float(ci))
    x = y = Decimal(0)
    k = 0
    margin = Decimal(10)
    while k < cap:
        r2 = x * x + y * y
        margin = min(margin, abs(r2 - 4))
        if r2 > 4:
            break
        x, y = x * x - y * y + cr, 2 * x * y + ci
        k += 1
    return k, margin


def test_sampled_pixels_match_high_precision():
    """Pixels whose orbit escapes quickly and never grazes the threshold have the
    same count in float32 as in exact arithmetic (error < 4^6 * 2^-24 << margin)."""
    pos = mandelbrot_positions(1024, 768)
    idx = np.random.default_rng(3).choice(pos.size, 3000, replace=False)
    got = oracle.mandelbrot(pos[idx], 256)
    checked = 0
    for i, g in zip(idx, got):
        k, margin = _decimal_count(pos[i]["re"], pos[i]["im"], 256)
        if k <= 6 and margin > Decimal("0.01"):
            assert g == k, (i, g, k)
            checked += 1
    assert checked > 1000


def test_positions_exact_dyadic():
    pos = mandelbrot_positions(1024, 768)
    assert pos[0]["re"] == -2.5 and pos[0]["im"] == -1.5
    assert pos[1]["re"] - pos[0]["re"] == 2.0 ** -8
    assert pos[1024]["im"] - pos[0]["im"] == 2.0 ** -8
    assert pos[-1]["re"] == np.float32(1.5 - 2.0 ** -8)


def test_whole_image_golden(golden_dir):
    """Independent numpy-float32 evaluation recorded in SURVEY.md §8c-c8."""
    with open(os.path.join(golden_dir, "mandelbrot.json")) as fh:
        g = json.load(fh)
    for case in g["cases"]:
        if case["width"] > 1024 or case["cap"] > 256:
            continue  # larger cases are checked in the slow test below
        pos = mandelbrot_positions(case["width"], case["height"])
        out = oracle.mandelbrot(pos, case["cap"])
        assert int(out.astype(np.int64).sum()) == case["sum_iter"]
        if "at_cap" in case:
            assert int((out == case["cap"]).sum()) == case["at_cap"]
        assert zlib.crc32(out.tobytes()) == int(case["crc32"], 16)


@pytest.mark.slow
def test_whole_image_golden_large(golden_dir):
    with open(os.path.join(golden_dir, "mandelbrot.json")) as fh:
        g = json.load(fh)
    for case in g["cases"]:
        if case["width"] <= 1024 and case["cap"] <= 256:
            continue
        pos = mandelbrot_positions(case["width"], case["height"])
        out = oracle.mandelbrot(pos, case["cap"])
        assert int(out.astype(np.int64).sum()) == case["sum_iter"]
        assert zlib.crc32(out.tobytes()) == int(case["crc32"], 16)


def test_golden_generator_reproduces_the_small_pin(golden_dir):
    """tests/golden/make_mandelbrot.py (numpy float32, independent of oracle/)
    regenerates the stored 1024x768@256 pin (the larger cases: run the script)."""
    import importlib.util
    spec = importlib.util.spec_from_file_location("make_mandelbrot",
                                                  os.path.join(golden_dir, "make_mandelbrot.py"))
    mk = importlib.util.module_from_spec(spec)
    spec.loader.exec_module(mk)
    with open(os.path.join(golden_dir, "mandelbrot.json")) as fh:
        want = json.load(fh)["cases"][0]
    assert mk.pins(want["width"], want["height"], want["cap"]) == want


def test_cyclic_rows_balance_the_devices():
    """NEXT-4: work per device (the oracle's iteration counts summed over the
    rows each device computes) for the paper's image (4096x3072, cap 256).
    Block rows: the busiest device carries 1.997 / 2.115 / 3.112x
    the mean at D = 2 / 4 / 8 (SURVEY §8d config 3's ideal-speedup ceiling).
    Cyclic rows (device k: rows k, k+D, ...): every device within 5% of the
    busiest (mean/max >= 0.95)."""
    W, H = 4096, 3072
    rows = oracle.mandelbrot(mandelbrot_positions(W, H), 256).astype(np.int64).reshape(H, W).sum(axis=1)
    total = rows.sum()
    for D, ceiling in ((2, 1.997), (3, None), (4, 2.115), (8, 3.112)):
        R = -(-H // D)
        block = np.array([rows[k * R:(k + 1) * R].sum() for k in range(D)])
        if ceiling is not None:
            assert abs(total / block.max() - ceiling) < 0.002, (D, total / block.max())
        cyc = np.array([rows[k::D].sum() for k in range(D)])
        assert cyc.sum() == total
        assert cyc.mean() / cyc.max() >= 0.95, (D, cyc.mean() / cyc.max())
