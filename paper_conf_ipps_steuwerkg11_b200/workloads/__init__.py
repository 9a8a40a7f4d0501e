"""Customizing functions (user source text) of the paper's workloads and of
the skeleton benchmarks.  They are *inputs* to the skeletons, handed to
libskel as strings and compiled by NVRTC into the skeleton
kernels."""
from pathlib import Path

_HERE = Path(__file__).resolve().parent


def source(name: str) -> str:
    return (_HERE / f"{name}.cu").read_text()


MANDELBROT = source("mandelbrot")
MANDELBROT_INDEX = source("mandelbrot_index")  # index Map variant (NEXT-4)
MANDELBROT_BLOCKED = source("mandelbrot_blocked")  # loop control per block of updates (NEXT-4)
# the blocked function with exact periodicity checking (a member is recognised
# when its float32 orbit repeats bit for bit; NEXT-4)
MANDELBROT_PERIODIC = "#define MANDEL_PERIODIC 1\n#define MANDEL_PRE 8\n" + MANDELBROT_BLOCKED
# 8 x 4 pixel tiles per warp: a void index Map writing the row-major image (NEXT-4)
MANDELBROT_TILES = MANDELBROT_BLOCKED + source("mandelbrot_tiles")
# the tiles with periodicity checking (coherent warps stop together: deep caps)
MANDELBROT_TILES_PERIODIC = "#define MANDEL_PERIODIC 1\n#define MANDEL_PRE 8\n" + MANDELBROT_TILES
# pairs of neighbouring pixels per element, packed FP32x2 arithmetic (NEXT-4)
MANDELBROT_PAIRS = source("mandelbrot_pairs")
# + exact periodicity checking, the pair kept in the packed loop until both
# pixels are done (no per-pixel finishing loops: MANDEL_NOREPLAY)
MANDELBROT_PAIRS_PERIODIC = "#define MANDEL_PERIODIC 1\n#define MANDEL_NOREPLAY 1\n" + MANDELBROT_PAIRS
# cyclic rows: index Map over a permuted row order (device k: rows k, k+D, ...),
# then an index Map that restores row-major order (NEXT-4; mandelbrot.py)
# (the pairs in their fastest form: lockstep packed loop with periodicity checking)
MANDELBROT_CYCLIC = MANDELBROT_PAIRS_PERIODIC + source("mandelbrot_cyclic")
MANDELBROT_UNPERMUTE = source("mandelbrot_unpermute")
# (the error-image Maps keep their direct event loads: SKEL_STAGE_ELEMS 0)
LMOSEM_ERROR = "#define SKEL_STAGE_ELEMS 0\n" + source("lmosem_error")
# the same function for prepared (longest-path-first) event order, where the
# Map is bound by L1TEX requests: 16-byte gathers per 4-float group in the
# forward projection too; in the given order they are slower
LMOSEM_ERROR_PREPARED = "#define LMOSEM_VEC_FWD 1\n" + LMOSEM_ERROR
# the same Listing 3 body on a lanes Map: `lanes` threads per event, each
# walking an alpha piece of the line of response (small per-GPU parts, §4.2)
LMOSEM_LANES = LMOSEM_ERROR + source("lmosem_lanes")
LMOSEM_LANES_PREPARED = "#define LMOSEM_VEC_FWD 1\n" + LMOSEM_LANES
LMOSEM_UPDATE = source("lmosem_update")
# FP32 lane-peak probe (measurement only: the Mandelbrot roofline's denominator)
PROBE_FP32 = source("probe_fp32")
PROBE_FP32_OPS_PER_STEP = 2 * 8  # FP32 operations per element and step (8 chains of add.rn.f32x2)
# on-device ordering of a subset's events by path length (Map + Scan + Map):
# bucket counts, then the scatter into bucket order (lmosem_order.cu)
_ORDER = source("lmosem_error") + source("lmosem_order")  # staged 24-byte event loads
LMOSEM_ORDER_HIST = _ORDER + """
void lm_order_hist(Event e, int *hist, int nx, int ny, int nz, int nb) {
    const int k = lm_slot(e, nx, ny, nz, nb);
    // lanes of a warp with the same counter add once
    const unsigned peers = __match_any_sync(__activemask(), k);
    if ((int)(threadIdx.x & 31u) == __ffs(peers) - 1) atomicAdd(&hist[k], __popc(peers));
}
"""
LMOSEM_ORDER_SCATTER = _ORDER + """
void lm_order_scatter(Event e, int *cursor, Event *out, int nx, int ny, int nz, int nb) {
    const int k = lm_slot(e, nx, ny, nz, nb);
    const unsigned peers = __match_any_sync(__activemask(), k);
    const int lane = (int)(threadIdx.x & 31u), leader = __ffs(peers) - 1;
    int base = 0;
    if (lane == leader) base = atomicAdd(&cursor[k], __popc(peers));
    base = __shfl_sync(peers, base, leader);
    out[base + __popc(peers & ((1u << lane) - 1u))] = e;
}
"""
LMOSEM_ORDER_BUCKETS = 64
LMOSEM_ORDER_REPLICAS = 128  # counters per bucket (lmosem_order.cu: lm_slot)
LMOSEM_ORDER_SLOTS = LMOSEM_ORDER_BUCKETS * LMOSEM_ORDER_REPLICAS * 8  # one counter per 32-byte sector
# voxel visits of one event's path (measurement only: the LM OSEM roofline
# counts one scattered request per visit in each of the two walks)
LMOSEM_VISITS = LMOSEM_ERROR + """
int lmosem_visits(Event e, int nx, int ny, int nz) {
    Walk w;
    if (!walk_init(e, nx, ny, nz, w)) return 0;
    return w.n_cross + 1;  // one segment per crossing, then the last one
}
"""
# 4-float groups the back projection reduces into (one red.global.add.v4.f32 each)
LMOSEM_GROUPS = LMOSEM_ERROR + """
static __forceinline__ void count_group(int v, float len, unsigned nvox, int &g, int &n) {
    if (len > 0.0f && (unsigned)v < nvox && (v >> 2) != g) {
        g = v >> 2;
        ++n;
    }
}
int lmosem_groups(Event e, int nx, int ny, int nz) {
    Walk w;
    if (!walk_init(e, nx, ny, nz, w)) return 0;
    Cursor cur;
    cursor_init(w, cur);
    int g = -1, n = 0;
    for (int it = 0; it < w.n_cross; ++it) {
        int vs;
        const double a1 = cross_step(w, cur, vs, true);
        count_group(vs, (float)((a1 - cur.ac) * w.len_scale), w.nvox, g, n);
        cur.ac = a1;
    }
    count_group(cur.v, (float)((w.amax - cur.ac) * w.len_scale), w.nvox, g, n);
    return n;
}
"""
PROBE_SCATTER_RED = source("probe_scatter")
PROBE_SCATTER_RED4 = source("probe_scatter4")
PROBE_GATHER = source("probe_gather")
PROBE_K = 64

# Listing 1, verbatim
SUM_F32 = "float sum (float x,float y){return x+y;}"
MULT_F32 = "float mult(float x,float y){return x*y;}"
SUM_I32 = "int sum(int x, int y){ return x + y; }"
# skeleton sweep
SAXPY_F32 = "float saxpy(float x, float y, float a){ return a * x + y; }"
SAXPY_I32 = "int saxpy(int x, int y, int a){ return a * x + y; }"
MAP_F32 = "float affine(float x){ return x * 2.0f + 1.0f; }"
MAP_I32 = "int affine(int x){ return x * 2 + 1; }"
