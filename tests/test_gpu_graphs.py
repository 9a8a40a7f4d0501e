"""CUDA-graph capture/replay of skeleton sequences (skel_capture_begin/end,
skel_graph_launch): replays must give exactly what eager execution gives,
including the Scan, whose look-back status words are tagged with a
device-resident epoch that every replay advances."""
import numpy as np
import pytest

import oracle
import skel_inputs as si
from paper_conf_ipps_steuwerkg11_b200 import skel
from paper_conf_ipps_steuwerkg11_b200.lmosem import LMOSEM
from paper_conf_ipps_steuwerkg11_b200.workloads import MAP_F32, SAXPY_F32, SUM_F32, SUM_I32

pytestmark = pytest.mark.gpu


@pytest.mark.parametrize("D", [1, 3])
def test_replayed_step_equals_eager(D):
    n = (1 << 21) + 5
    x, y = si.uniform_f32(n, 1), si.uniform_f32(n, 2)
    with skel.Context(D) as ctx:
        X, Y = ctx.vector(x), ctx.vector(y)
        if D > 1:
            X.set_distribution(skel.BLOCK)
        m, z, s = (ctx.vector(n=n, dtype=np.float32) for _ in range(3))
        r = ctx.vector(n=1, dtype=np.float32)

        def step():
            ctx.map(MAP_F32, X, m)
            ctx.zip(SAXPY_F32, X, Y, z, args=[np.float32(2.5)])
            ctx.reduce_to(SUM_F32, X, r)
            ctx.scan(SUM_F32, X, s, np.float32(0))

        step()  # eager warm-up: compiles, uploads, allocates
        want = [v.download() for v in (m, z, s, r)]
        for v in (m, z, s, r):
            v.fill(np.float32(-1))
        g = ctx.capture(step)
        for _ in range(4):
            g.launch()
        got = [v.download() for v in (m, z, s, r)]
        for a, b in zip(got, want):
            assert np.array_equal(a, b)
        g.destroy()


def test_scan_replays_see_new_data():
    """Scan statuses from the previous replay must never be taken as current."""
    n = 3 * 16384 * 148 + 999  # several slices and a ragged tail
    x = si.uniform_int01(n, 3)
    with skel.Context(1) as ctx:
        X = ctx.vector(x)
        out = ctx.vector(n=n, dtype=np.int32)
        ctx.scan(SUM_I32, X, out, np.int32(0))
        g = ctx.capture(lambda: ctx.scan(SUM_I32, X, out, np.int32(0)))
        inc = "int inc(int v){ return v + 1; }"
        ctx.prepare("map", inc)
        cur = x.copy()
        for _ in range(3):
            ctx.map(inc, X, X)  # eager: new input every round
            cur = cur + 1
            g.launch()
            assert np.array_equal(out.download(), oracle.skel_scan(SUM_I32, cur, 0))
        g.destroy()


def test_blocking_calls_rejected_while_capturing():
    with skel.Context(1) as ctx:
        v = ctx.vector(np.ones(10, np.float32))
        ctx.map(MAP_F32, v, v)
        ctx.capture_begin()
        with pytest.raises(skel.SkelError) as e:
            v.download()
        assert e.value.name == "SKEL_ERR_STATE"
        with pytest.raises(skel.SkelError) as e:
            ctx.map("float neverseen(float x){ return x; }", v, v)  # would compile
        assert e.value.name == "SKEL_ERR_STATE"
        ctx.capture_end().destroy()


@pytest.mark.parametrize("D", [1, 4])
def test_lmosem_subset_graph(D):
    ev = si.lmosem_events(20_000, subset=1)
    imgs = []
    for use_graph in (False, True):
        with skel.Context(D) as ctx:
            rec = LMOSEM(ctx)
            evv = rec.events(ev)
            rec.subset(evv)  # first subset eagerly (warm-up)
            if use_graph:
                g = ctx.capture(lambda: rec.subset(evv))
                g.launch()
                g.launch()
                g.destroy()
            else:
                rec.subset(evv)
                rec.subset(evv)
            imgs.append(rec.image())
    # same three subsets (atomic order may differ)
    a, b = (i.astype(np.float64) for i in imgs)
    assert np.linalg.norm(a - b) <= 1e-5 * np.linalg.norm(a)
