"""Lazy host/device coherence of Vector (§III-A), observed
through the library's transfer counters on the Listing 1 pattern."""
import numpy as np
import pytest

import oracle
import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.workloads import MAP_F32, MULT_F32, SUM_F32

pytestmark = pytest.mark.gpu


def test_listing1_transfers():
    n = 1 << 18
    a, b = si.uniform_f32(n, 1), si.uniform_f32(n, 2)
    with skel.Context(1) as ctx:
        A, B = ctx.vector(a), ctx.vector(b)
        ctx.prepare("zip", MULT_F32)
        ctx.prepare("reduce", SUM_F32)
        ctx.reset_stats()
        st = ctx.stats()
        assert st["h2d_bytes"] == 0  # upload only fills the host mirror (lazy)
        prod = ctx.vector(n=n, dtype=np.float32)
        ctx.zip(MULT_F32, A, B, prod)
        st = ctx.stats()
        assert st["h2d_copies"] == 2 and st["h2d_bytes"] == 2 * n * 4  # one H2D per input
        c = ctx.reduce(SUM_F32, prod)
        st = ctx.stats()
        assert st["d2h_copies"] == 1 and st["d2h_bytes"] == 4  # only the scalar comes back
        # the intermediate never travelled; the result matches
        want = oracle.sum_f32_exact(oracle.skel_zip(MULT_F32, a, b, np.float32))
        assert abs(float(c) - want) <= 1e-5 * abs(want)
        # a second skeleton on the same inputs transfers nothing
        ctx.zip(MULT_F32, A, B, prod)
        assert ctx.stats()["h2d_bytes"] == 2 * n * 4


def test_download_only_when_devices_are_newer():
    x = si.uniform_f32(10_000, 3)
    with skel.Context(1) as ctx:
        v = ctx.vector(x)
        ctx.reset_stats()
        assert np.array_equal(v.download(), x)  # host copy valid: no D2H
        assert ctx.stats()["d2h_bytes"] == 0
        out = ctx.vector(n=x.size, dtype=np.float32)
        ctx.map(MAP_F32, v, out)
        r1 = out.download()
        r2 = out.download()
        assert ctx.stats()["d2h_copies"] == 1  # second download is served from the host copy
        assert np.array_equal(r1, r2)


def test_host_write_after_device_write_reuploads():
    x = si.uniform_f32(5000, 4)
    with skel.Context(1) as ctx:
        v = ctx.vector(x)
        out = ctx.vector(n=x.size, dtype=np.float32)
        ctx.map(MAP_F32, v, v)  # device copy is newer now
        y = x + 1
        v.upload(y)  # host write: next skeleton must re-upload
        ctx.reset_stats()
        ctx.map(MAP_F32, v, out)
        assert ctx.stats()["h2d_bytes"] == x.size * 4
        assert np.array_equal(out.download(), oracle.skel_map(MAP_F32, y.astype(np.float32), np.float32))


def test_host_view_zero_copy_write():
    x = si.uniform_f32(4096, 5)
    with skel.Context(1) as ctx:
        v = ctx.vector(n=x.size, dtype=np.float32)
        hv = v.host_view()
        hv[:] = x
        v.mark_host_modified()
        out = ctx.vector(n=x.size, dtype=np.float32)
        ctx.map(MAP_F32, v, out)
        assert np.array_equal(out.download(), oracle.skel_map(MAP_F32, x, np.float32))


def test_create_is_zero_filled_and_fill():
    with skel.Context(1) as ctx:
        v = ctx.vector(n=1000, dtype=np.float32)
        assert not v.download().any()
        v.fill(np.float32(2.5))
        assert (v.download() == 2.5).all()


def test_disk_kernel_cache_roundtrip(tmp_path):
    """compiled kernels are saved on disk and loaded later."""
    src = "float plus7(float x){ return x + 7.0f; }"
    with skel.Context(1) as ctx:
        ctx.set_cache_dir(str(tmp_path))
        ctx.prepare("map", src)
        s = ctx.stats()
        assert s["compile_misses"] == 1
    assert any(p.suffix == ".cubin" for p in tmp_path.iterdir())
    with skel.Context(1) as ctx:
        ctx.set_cache_dir(str(tmp_path))
        x = np.arange(10, dtype=np.float32)
        out = ctx.vector(n=10, dtype=np.float32)
        ctx.map(src, ctx.vector(x), out)
        s = ctx.stats()
        assert s["compile_disk_hits"] == 1 and s["compile_misses"] == 0
        assert np.array_equal(out.download(), x + 7)


@pytest.mark.parametrize("D", [1, 4])
@pytest.mark.parametrize("dist", ["single", "block", "copy"])
def test_download_part_reads_the_range_from_the_devices(D, dist):
    """download_part (the counterpart of upload_part): a range comes
    straight from the device storage that holds it -- exactly its bytes, no
    full-vector D2H, the host mirror untouched -- and from the host mirror when
    that is valid."""
    n = 100_003
    x = si.uniform_f32(n, 7)
    with skel.Context(D) as ctx:
        v = ctx.vector(x)
        out = ctx.vector(n=n, dtype=np.float32)
        v.set_distribution({"single": skel.SINGLE, "block": skel.BLOCK, "copy": skel.COPY}[dist])
        ctx.map(MAP_F32, v, out)
        want = oracle.skel_map(MAP_F32, x, np.float32)
        ctx.sync()
        ctx.reset_stats()
        for lo, cnt in ((0, n), (0, 1), (n - 1, 1), (25_000, 50_001), (12_345, 0)):
            got = out.download_part(lo, np.empty(cnt, np.float32))
            assert np.array_equal(got, want[lo:lo + cnt])
        st = ctx.stats()
        assert st["d2h_bytes"] == 4 * (n + 1 + 1 + 50_001)  # only the ranges travelled
        # a full download validates the mirror; a later part is a host memcpy
        assert np.array_equal(out.download(), want)
        ctx.reset_stats()
        assert np.array_equal(out.download_part(3, np.empty(10, np.float32)), want[3:13])
        assert ctx.stats()["d2h_bytes"] == 0
        with pytest.raises(skel.SkelError) as e:
            out.download_part(n - 2, np.empty(3, np.float32))
        assert e.value.name == "SKEL_ERR_SIZE"


def test_download_part_async_overlaps_and_orders_writes():
    """skel_vector_download_part_async: the copy is enqueued on the download
    stream after everything already enqueued for the vector; a later skeleton
    that rewrites the vector waits for it on the device (write-after-read), so
    the host buffer holds the values as of the call; skel_sync completes it."""
    import torch
    n = (1 << 22) + 3
    x = si.uniform_f32(n, 12)
    with skel.Context(1) as ctx:
        v = ctx.vector(x)
        out = ctx.vector(n=n, dtype=np.float32)
        ctx.map(MAP_F32, v, out)
        host = torch.empty(n, dtype=torch.float32, pin_memory=True).numpy()
        out.download_part_async(0, host)
        for _ in range(5):  # rewrite out in place right away: must not race the copy
            ctx.map(MAP_F32, out, out)
        ctx.sync()
        want = oracle.skel_map(MAP_F32, x, np.float32)
        assert np.array_equal(host, want)
        w = want
        for _ in range(5):
            w = oracle.skel_map(MAP_F32, w, np.float32)
        assert np.array_equal(out.download(), w)
        part = torch.empty(1000, dtype=torch.float32, pin_memory=True).numpy()
        out.download_part_async(n - 1000, part)
        ctx.sync()
        assert np.array_equal(part, w[-1000:])


@pytest.mark.parametrize("D", [3, 4])
def test_download_part_async_block_parts_on_virtual_devices(D):
    """download_part_async of a range spanning several devices' block parts:
    one D2H per overlapping part on each device's download stream."""
    import torch
    n = 1_000_003
    x = si.uniform_f32(n, 14)
    with skel.Context(D) as ctx:
        v = ctx.vector(x)
        v.set_distribution(skel.BLOCK)
        out = ctx.vector(n=n, dtype=np.float32)
        ctx.map(MAP_F32, v, out)
        lo, cnt = n // 7, n // 2
        host = torch.empty(cnt, dtype=torch.float32, pin_memory=True).numpy()
        ctx.reset_stats()
        out.download_part_async(lo, host)
        ctx.map(MAP_F32, out, out)  # waits for the copies on every device
        ctx.sync()
        assert ctx.stats()["d2h_bytes"] == 4 * cnt
        want = oracle.skel_map(MAP_F32, x, np.float32)
        assert np.array_equal(host, want[lo:lo + cnt])
        assert np.array_equal(out.download(), oracle.skel_map(MAP_F32, want, np.float32))
