"""GPU parity of the Mandelbrot Map (§IV-A, eq. (5)): bit-exact
iteration counts against the oracle and the golden whole-image pins, on one
device and block-distributed over virtual devices (rows split)."""
import json
import os
import zlib

import numpy as np
import pytest

import oracle
import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import MANDELBROT

pytestmark = pytest.mark.gpu


def run(ctx, pos, cap, dist=None, fn=MANDELBROT):
    vin = ctx.vector(pos)
    if dist is not None:
        vin.set_distribution(dist)
    out = ctx.vector(n=pos.size, dtype=np.int32)
    ctx.map(fn, vin, out, args=[np.int32(cap)])
    return out.download()


def test_closed_form_points():
    cs = [1 + 0j, 2 + 0j, -1.5 + 1.5j, 0j, -1 + 0j, -2 + 0j, 1j, 0.25 + 0j, 3 + 0j]
    want = [3, 2, 1, 256, 256, 256, 256, 256, 1]
    pos = np.zeros(len(cs), si.POS_DTYPE)
    pos["re"] = [c.real for c in cs]
    pos["im"] = [c.imag for c in cs]
    with skel.Context(1) as ctx:
        assert run(ctx, pos, 256).tolist() == want


@pytest.mark.parametrize("w,h,cap", [(1024, 768, 256), (4096, 3072, 256), (1024, 768, 4096)])
def test_whole_image_bit_exact(golden_dir, w, h, cap):
    pos = si.mandelbrot_positions(w, h)
    with skel.Context(1) as ctx:
        got = run(ctx, pos, cap)
    with open(os.path.join(golden_dir, "mandelbrot.json")) as fh:
        case = [c for c in json.load(fh)["cases"] if (c["width"], c["height"], c["cap"]) == (w, h, cap)][0]
    assert zlib.crc32(got.tobytes()) == int(case["crc32"], 16)
    assert int(got.astype(np.int64).sum()) == case["sum_iter"]
    if w * h <= 1 << 20:
        assert np.array_equal(got, oracle.mandelbrot(pos, cap))


@pytest.mark.parametrize("D", [2, 3, 4, 8])
def test_block_rows_on_virtual_devices(D):
    pos = si.mandelbrot_positions(1024, 768)
    with skel.Context(D) as ctx:
        got = run(ctx, pos, 256, skel.BLOCK)
    assert np.array_equal(got, oracle.mandelbrot(pos, 256))


@pytest.mark.parametrize("w,h,cap,D", [(1024, 768, 256, 1), (4096, 3072, 256, 1), (1024, 768, 256, 3)])
def test_index_map_variant_matches_the_golden_image(golden_dir, w, h, cap, D):
    """NEXT-4: the same image from an index Map (c computed in the kernel from
    the pixel index, no position vector) -- bit-identical to the golden pins."""
    from paper_conf_ipps_steuwerkg11_b200.workloads import MANDELBROT_INDEX
    with skel.Context(D) as ctx:
        out = ctx.vector(n=w * h, dtype=np.int32)
        if D > 1:
            out.set_distribution(skel.BLOCK)
        ctx.map_index(MANDELBROT_INDEX, w * h, out, args=[np.int32(w), np.int32(h), np.int32(cap)])
        got = out.download()
    with open(os.path.join(golden_dir, "mandelbrot.json")) as fh:
        case = [c for c in json.load(fh)["cases"] if (c["width"], c["height"], c["cap"]) == (w, h, cap)][0]
    assert zlib.crc32(got.tobytes()) == int(case["crc32"], 16)


@pytest.mark.parametrize("w,h,cap,D", [(1024, 768, 256, 1), (4096, 3072, 256, 1), (1024, 768, 4096, 1),
                                       (1024, 768, 256, 4), (257, 3, 9, 1)])
def test_blocked_variant_bit_exact(golden_dir, w, h, cap, D):
    """NEXT-4: the blocked user function (loop control per 8 updates, roll back
    on escape) gives the same counts as eq. (5) as written: golden CRCs and the
    oracle, on one device and block-distributed rows; a ragged 257x3 image with
    a cap that is not a multiple of the block."""
    from paper_conf_ipps_steuwerkg11_b200.workloads import MANDELBROT_BLOCKED
    pos = si.mandelbrot_positions(w, h)
    with skel.Context(D) as ctx:
        got = run(ctx, pos, cap, skel.BLOCK if D > 1 else None, fn=MANDELBROT_BLOCKED)
    cases = json.load(open(os.path.join(golden_dir, "mandelbrot.json")))["cases"]
    case = [c for c in cases if (c["width"], c["height"], c["cap"]) == (w, h, cap)]
    if case:
        assert zlib.crc32(got.tobytes()) == int(case[0]["crc32"], 16)
    if w * h <= 1 << 20:
        assert np.array_equal(got, oracle.mandelbrot(pos, cap))


@pytest.mark.parametrize("w,h,cap,D", [(1024, 768, 256, 1), (4096, 3072, 256, 1), (1024, 768, 4096, 1),
                                       (1024, 768, 256, 4), (1024, 768, 7, 1), (1024, 768, 1500, 1)])
def test_pairs_variant_bit_exact(golden_dir, w, h, cap, D):
    """mandelbrot_pairs.cu (two neighbouring pixels per element, packed FFMA2 /
    FADD2 arithmetic with the multiplies kept unfused): the same counts as eq.
    (5) as written -- golden CRCs and the oracle, on one and on four devices."""
    from paper_conf_ipps_steuwerkg11_b200.workloads import MANDELBROT_PAIRS, MANDELBROT_PAIRS_PERIODIC
    pos = si.mandelbrot_positions(w, h)
    pairs = pos.view(si.POS2_DTYPE)
    for fn in (MANDELBROT_PAIRS, MANDELBROT_PAIRS_PERIODIC):
        _pairs_check(golden_dir, w, h, cap, D, pos, pairs, fn)


def _pairs_check(golden_dir, w, h, cap, D, pos, pairs, MANDELBROT_PAIRS):
    with skel.Context(D) as ctx:
        vin = ctx.vector(pairs)
        if D > 1:
            vin.set_distribution(skel.BLOCK)
        out = ctx.vector(n=pairs.size, dtype=si.CNT2_DTYPE)
        ctx.map(MANDELBROT_PAIRS, vin, out, args=[np.int32(cap)])
        got = out.download().view(np.int32)
    with open(os.path.join(golden_dir, "mandelbrot.json")) as fh:
        cases = [c for c in json.load(fh)["cases"] if (c["width"], c["height"], c["cap"]) == (w, h, cap)]
    if cases:
        assert zlib.crc32(got.tobytes()) == int(cases[0]["crc32"], 16)
    if w * h <= 1 << 20:
        assert np.array_equal(got, oracle.mandelbrot(pos, cap))


@pytest.mark.parametrize("w,h,cap,D", [(1024, 768, 256, 1), (1024, 768, 256, 2), (1024, 768, 256, 3),
                                       (1024, 768, 256, 4), (1024, 768, 256, 8), (4096, 3072, 256, 8),
                                       (1024, 768, 4096, 4), (258, 7, 50, 3)])
def test_cyclic_rows_bit_exact(golden_dir, w, h, cap, D):
    """NEXT-4 cyclic rows (mandelbrot.CyclicMandelbrot): device k computes rows
    k, k+D, ... into a permuted, block-distributed image; gathered and
    un-permuted on device 0 it is the golden image (and the oracle's), also
    when the rows do not divide evenly (258x7 at D = 3: padding slots)."""
    from paper_conf_ipps_steuwerkg11_b200.mandelbrot import CyclicMandelbrot
    with skel.Context(D) as ctx:
        cm = CyclicMandelbrot(ctx, w, h)
        got = cm.counts(cap)
        again = cm.counts(cap)  # buffers reused
    assert np.array_equal(got, again)
    cases = [c for c in json.load(open(os.path.join(golden_dir, "mandelbrot.json")))["cases"]
             if (c["width"], c["height"], c["cap"]) == (w, h, cap)]
    if cases:
        assert zlib.crc32(got.tobytes()) == int(cases[0]["crc32"], 16)
    if w * h <= 1 << 20:
        assert np.array_equal(got, oracle.mandelbrot(si.mandelbrot_positions(w, h), cap))


@pytest.mark.parametrize("w,h,cap,D", [(1024, 768, 256, 1), (4096, 3072, 256, 1), (1024, 768, 4096, 1),
                                       (1024, 768, 256, 3)])
def test_tiles_variant_bit_exact(golden_dir, w, h, cap, D):
    """NEXT-4: 8 x 4 pixel tiles per warp (void index Map writing the row-major
    image through a vector argument): the golden image."""
    from paper_conf_ipps_steuwerkg11_b200.workloads import MANDELBROT_TILES
    with skel.Context(D) as ctx:
        img = ctx.vector(n=w * h, dtype=np.int32)
        img.fill_dist(skel.COPY if D > 1 else skel.SINGLE, np.int32(-1))
        ctx.map_index(MANDELBROT_TILES, w * h, None, args=[img, np.int32(w), np.int32(h), np.int32(cap)])
        img.mark_device_modified()
        if D > 1:  # each device wrote its own tiles into its copy: combine (max over -1 fill)
            img.set_distribution(skel.SINGLE, skel.COMBINE_MAX)
        got = img.download()
    cases = [c for c in json.load(open(os.path.join(golden_dir, "mandelbrot.json")))["cases"]
             if (c["width"], c["height"], c["cap"]) == (w, h, cap)]
    assert zlib.crc32(got.tobytes()) == int(cases[0]["crc32"], 16)


@pytest.mark.parametrize("w,h,cap,D", [(1024, 768, 256, 1), (4096, 3072, 256, 1), (1024, 768, 4096, 1),
                                       (1024, 768, 256, 4), (257, 3, 9, 1)])
def test_periodic_variant_bit_exact(golden_dir, w, h, cap, D):
    """NEXT-4: the blocked function with exact periodicity checking (a member
    recognised when its float32 orbit repeats bit for bit): the counts of eq.
    (5) as written -- golden CRCs and the oracle."""
    from paper_conf_ipps_steuwerkg11_b200.workloads import MANDELBROT_PERIODIC
    pos = si.mandelbrot_positions(w, h)
    with skel.Context(D) as ctx:
        got = run(ctx, pos, cap, skel.BLOCK if D > 1 else None, fn=MANDELBROT_PERIODIC)
    cases = [c for c in json.load(open(os.path.join(golden_dir, "mandelbrot.json")))["cases"]
             if (c["width"], c["height"], c["cap"]) == (w, h, cap)]
    if cases:
        assert zlib.crc32(got.tobytes()) == int(cases[0]["crc32"], 16)
    if w * h <= 1 << 20:
        assert np.array_equal(got, oracle.mandelbrot(pos, cap))


@pytest.mark.parametrize("w,h,cap", [(1024, 768, 256), (1024, 768, 4096), (4096, 3072, 256)])
def test_tiles_periodic_variant_bit_exact(golden_dir, w, h, cap):
    from paper_conf_ipps_steuwerkg11_b200.workloads import MANDELBROT_TILES_PERIODIC
    with skel.Context(1) as ctx:
        img = ctx.vector(n=w * h, dtype=np.int32)
        ctx.map_index(MANDELBROT_TILES_PERIODIC, w * h, None, args=[img, np.int32(w), np.int32(h), np.int32(cap)])
        img.mark_device_modified()
        got = img.download()
    cases = [c for c in json.load(open(os.path.join(golden_dir, "mandelbrot.json")))["cases"]
             if (c["width"], c["height"], c["cap"]) == (w, h, cap)]
    assert zlib.crc32(got.tobytes()) == int(cases[0]["crc32"], 16)
