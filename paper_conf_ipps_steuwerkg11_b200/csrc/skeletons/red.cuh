// red.cuh -- Reduce (eq. (3)) and Scan (eq. (4))
// skeleton kernels for a user operator  T SKEL_FN(T x, T y, args...).
//
// (+) must be associative but need not be commutative, so
// every combination below keeps index order: the left operand always covers
// lower indices.  No identity is assumed for Reduce (eq. (3) has none);
// partial results carry a validity bit instead.
//
// B200 mapping (kernels K3/K4):
//  * A tile is RB = 512 threads x K elements, K*sizeof(T) = 128 bytes, i.e.
//    one 128-byte row per thread, 64 KB per tile.  Tiles are moved by the
//    TMA engine (cp.async.bulk.tensor.2d, 128B swizzle) into a 3-stage
//    shared-memory ring guarded by mbarriers; the swizzle lets each thread
//    read its own contiguous row with conflict-free 128-bit LDS (chunk j of
//    row r lives at chunk j ^ (r & 7)).  One CTA per SM.
//  * Reduce: static contiguous tile ranges per CTA, per-tile ordered block
//    reduction (in-thread fold, shuffle tree lower-lane-left, warps in
//    order), a running CTA aggregate, and a last-CTA-done ordered fold of the
//    CTA partials: a single pass over the input (4 B/element for float).
//  * Scan: a persistent grid (one CTA per SM, launched cooperatively so the
//    whole grid is co-resident) walks the vector in slices of G tiles; a
//    CTA publishes its tile aggregate A(s,c) and folds the window of G-1
//    aggregates W(s) = A(s-1,c+1..G-1) (+) A(s,0..c-1) ahead of its consumers
//    (the window waits on higher-index CTAs of the previous slice, hence the
//    co-residency requirement).  Status words carry an epoch so no memset is
//    needed between launches; outputs are staged in the same swizzled smem
//    stage and written by TMA tensor stores (8 B/element).
//  * Element types whose size is not 4, 8 or 16 bytes, unaligned views and
//    the ragged last tile use direct (LDG/STG) loads with the same ordering.
//  * A block-distributed Reduce over in-process devices ends inside these
//    kernels: the last device to finish folds the device results in device
//    order (skel_xdev_finish, system-scope ticket).
//  * The kernels are launched as programmatic dependents of the previous
//    kernel on the stream and wait for it first (griddepcontrol, prelude.cuh).

// Reduce main loop: 1 = direct 128-bit loads, every warp folding its own
// contiguous range (no barrier in the loop); 0 = TMA tiles through shared
// memory with one ordered block fold per tile (K3)
#ifndef SKEL_RED_DIRECT
#define SKEL_RED_DIRECT 0
#endif
#ifndef SKEL_RBLOCK
#if SKEL_RED_DIRECT
#define SKEL_RBLOCK 256
#else
#define SKEL_RBLOCK 512
#endif
#endif
#ifndef SKEL_RED_U
#define SKEL_RED_U 4  // direct Reduce: 16-byte loads in flight per lane
#endif
#ifndef SKEL_STAGES
#define SKEL_STAGES 3
#endif

using skel_F = decltype(&SKEL_FN);
using skel_FT = skel::fn<skel_F>;
using skel_T = skel::decay_t<typename skel_FT::ret>;
static_assert(skel_FT::arity >= 2, "Reduce/Scan need a binary operator");
static_assert(skel::same<typename skel_FT::template param<0>, skel_T>::value &&
                  skel::same<typename skel_FT::template param<1>, skel_T>::value,
              "Reduce/Scan operator must have the form T f(T, T, ...)");
using skel_Args = typename skel::drop<2, typename skel_FT::params>::type;
using skel_Lay = skel::args_layout<skel_Args>;
constexpr skel_u64 SKEL_ARGBYTES = skel::cmax<skel_u64>(16, skel::align_up(skel_Lay::bytes, 16));
using skel_Buf = skel::argbuf<SKEL_ARGBYTES>;
using skel_Seq = typename skel::make_iseq<skel_Lay::n>::type;
using skel_S = skel::slot<skel_T>;

constexpr int RB = SKEL_RBLOCK;
constexpr int NW = RB / 32;
constexpr bool TMA_OK = sizeof(skel_T) == 4 || sizeof(skel_T) == 8 || sizeof(skel_T) == 16;
constexpr int K = TMA_OK ? (int)(128 / sizeof(skel_T)) : (int)skel::cmax<skel_u64>(1, 128 / sizeof(skel_T));
constexpr bool RDIRECT = SKEL_RED_DIRECT != 0;
constexpr int RU = SKEL_RED_U;
constexpr int PERV = TMA_OK ? (int)(16 / sizeof(skel_T)) : 1;  // elements per 16-byte lane load
// Reduce work unit (elements): a TMA tile, or one round of RU loads of every warp
constexpr skel_u64 TILE = RDIRECT ? (skel_u64)RB * PERV * RU : (skel_u64)RB * K;
constexpr unsigned TILE_BYTES = (unsigned)((skel_u64)RB * K * sizeof(skel_T));
constexpr int STAGES = SKEL_STAGES;
// Reduce tile order: 0 = static contiguous tile ranges per CTA (one partial per
// CTA); 1 = tile i on CTA i mod G (all CTAs stream adjacent tiles, like a
// grid-stride loop), one partial per tile, folded in index order at the end
#ifndef SKEL_RED_INTERLEAVE
#define SKEL_RED_INTERLEAVE 0
#endif
constexpr bool RIL = SKEL_RED_INTERLEAVE != 0;
constexpr unsigned DSMEM = (TMA_OK && !RDIRECT) ? STAGES * TILE_BYTES + 1024 : 0;
// Scan: tiles per CTA per slice (see the Scan section)
#ifndef SKEL_SCAN_CH
#define SKEL_SCAN_CH 1
#endif
constexpr int SCAN_CH = SKEL_SCAN_CH;
#ifndef SKEL_SCAN_PW
#define SKEL_SCAN_PW 1
#endif
constexpr int PW = SKEL_SCAN_PW;  // Scan window warps (slices folded concurrently)
#ifndef SKEL_SCAN_RB
#define SKEL_SCAN_RB 512
#endif
#ifndef SKEL_SCAN_SPER
#define SKEL_SCAN_SPER 8  // small-vector Scan: elements per thread (tile = RB x SPER)
#endif
#ifndef SKEL_SCAN_STAGES
#define SKEL_SCAN_STAGES 3
#endif
constexpr int SRB = SKEL_SCAN_RB;  // consumer threads = rows per scan tile
constexpr int SNW = SRB / 32;
constexpr int SSTAGES = SKEL_SCAN_STAGES;
constexpr skel_u64 STILE = (skel_u64)SRB * K;
constexpr unsigned STILE_BYTES = (unsigned)(STILE * sizeof(skel_T));
constexpr unsigned SDSMEM = TMA_OK ? SSTAGES * STILE_BYTES + 1024 : 0;
constexpr bool PACKED = sizeof(skel_S) == 4;  // status = value:32 | epoch:30 | state:2
#ifndef SKEL_SCAN_REPL
#define SKEL_SCAN_REPL 8
#endif
// copies of every packed status word: CTA c polls copy c % REPL, so the few L2
// lines a slice's status occupies are not hammered by all G CTAs at once
// (2 copies measured 0.4% faster alone at 2^30 but slower inside the bench's
// sweep at 2^24..2^30, profiles/r01_bench_s4_repl2.json: 8 kept)
constexpr int REPL = PACKED ? SKEL_SCAN_REPL : 1;

struct skel_sig_t { skel_u64 v[16 + 4 * 32]; };
constexpr skel_sig_t skel_make_sig() {
    skel_sig_t s{};
    s.v[0] = 1;
    s.v[1] = 3;  // reduce/scan module
    s.v[2] = skel_FT::arity;
    s.v[3] = sizeof(skel_T);
    s.v[4] = sizeof(skel_S);
    s.v[5] = TMA_OK;
    s.v[6] = skel_Lay::n;
    s.v[7] = SKEL_ARGBYTES;
    s.v[8] = K;
    s.v[9] = RB;
    s.v[10] = TILE;
    s.v[11] = DSMEM;
    s.v[12] = SDSMEM;
    s.v[13] = PACKED;
    s.v[14] = SRB + 64 + 32 * PW;  // scan block size (consumers, producer, store and window warps); tile = SRB * K
    s.v[15] = (skel_u64)SRB | ((skel_u64)SCAN_CH << 16) | ((skel_u64)REPL << 32) |
              ((skel_u64)RIL << 48) | ((skel_u64)RDIRECT << 49) | ((skel_u64)SKEL_SCAN_SPER << 50);  // scan rows/tile | tiles/CTA/slice | status
                                                                  // copies | reduce tile order | direct reduce
    for (int i = 0; i < skel_Lay::n && i < 32; ++i) {
        s.v[16 + 4 * i] = skel_Lay::size(i);
        s.v[17 + 4 * i] = skel_Lay::align(i);
        s.v[18 + 4 * i] = skel_Lay::isptr(i);
        s.v[19 + 4 * i] = skel_Lay::off(i);
    }
    return s;
}
extern "C" __device__ skel_sig_t skel_sig = skel_make_sig();

struct skel_tmap { alignas(64) skel_u64 w[16]; };  // CUtensorMap (opaque, 128 B)

// (valid, value) pair: a partial result over a possibly empty index range
struct VT {
    skel_T v;
    bool ok;
};

template <class Tup> __device__ __forceinline__ skel_T opf(const skel_T &a, const skel_T &b, Tup &t) {
    return skel::caller<skel_Seq>::call(&SKEL_FN, t, a, b);
}
// a covers lower indices than b
template <class Tup> __device__ __forceinline__ VT comb(const VT &a, const VT &b, Tup &t) {
    if (!a.ok) return b;
    if (!b.ok) return a;
    VT r;
    r.v = opf(a.v, b.v, t);
    r.ok = true;
    return r;
}
__device__ __forceinline__ VT vt_shfl_down(const VT &x, int d) {
    VT r;
    r.v = skel::shfl_down(x.v, d);
    r.ok = __shfl_down_sync(0xffffffffu, (int)x.ok, d) != 0;
    return r;
}
__device__ __forceinline__ VT vt_shfl_up(const VT &x, int d) {
    VT r;
    r.v = skel::shfl_up(x.v, d);
    r.ok = __shfl_up_sync(0xffffffffu, (int)x.ok, d) != 0;
    return r;
}
__device__ __forceinline__ VT vt_shfl_idx(const VT &x, int s) {
    VT r;
    r.v = skel::shfl_idx(x.v, s);
    r.ok = __shfl_sync(0xffffffffu, (int)x.ok, s) != 0;
    return r;
}

// ordered warp fold: lane 0 receives x_0 (+) x_1 (+) ... (+) x_31
template <class Tup> __device__ __forceinline__ VT warp_fold(VT x, int lane, Tup &t) {
#pragma unroll
    for (int d = 1; d < 32; d <<= 1) {
        VT o = vt_shfl_down(x, d);
        if ((lane & (2 * d - 1)) == 0) x = comb(x, o, t);
    }
    return x;
}
// ordered block fold; result valid in thread 0.  Uses wpart[NW] + 1 barrier.
template <class Tup> __device__ __forceinline__ VT block_fold(VT x, VT *wpart, Tup &t) {
    const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
    x = warp_fold(x, lane, t);
    if (lane == 0) wpart[w] = x;
    __syncthreads();
    VT r;
    r.ok = false;
    if (w == 0) {
        VT y;
        y.ok = false;
        if (lane < NW) y = wpart[lane];
        r = warp_fold(y, lane, t);
    }
    return r;
}
// ordered block exclusive scan of per-thread values; returns the exclusive
// prefix of this thread (ok == false for an empty prefix) and writes the
// block total to *total.  Uses wsc[NW] + 2 barriers.
template <class Tup> __device__ __forceinline__ VT block_exscan(VT x, VT *wsc, VT *total, Tup &t) {
    const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
    VT inc = x;
#pragma unroll
    for (int d = 1; d < 32; d <<= 1) {
        VT o = vt_shfl_up(inc, d);
        if (lane >= d) inc = comb(o, inc, t);
    }
    VT ex = vt_shfl_up(inc, 1);
    if (lane == 0) ex.ok = false;
    if (lane == 31) wsc[w] = inc;
    __syncthreads();
    if (w == 0) {
        VT y;
        y.ok = false;
        if (lane < NW) y = wsc[lane];
        VT yi = y;
#pragma unroll
        for (int d = 1; d < 32; d <<= 1) {
            VT o = vt_shfl_up(yi, d);
            if (lane >= d) yi = comb(o, yi, t);
        }
        VT ye = vt_shfl_up(yi, 1);
        if (lane == 0) ye.ok = false;
        if (lane < NW) wsc[lane] = ye;
        if (lane == NW - 1) *total = yi;
    }
    __syncthreads();
    return comb(wsc[w], ex, t);
}

// ---- TMA helpers -----------------------------------------------------------
__device__ __forceinline__ void tma_load_rows(void *dst, const skel_tmap *map, int row, skel_u64 *bar) {
    asm volatile(
        "cp.async.bulk.tensor.2d.shared::cluster.global.tile.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3}], [%4];" ::"r"(
            skel::smem_addr(dst)),
        "l"(map), "r"(0), "r"(row), "r"(skel::smem_addr(bar))
        : "memory");
}
__device__ __forceinline__ void tma_store_rows(const skel_tmap *map, int row, const void *src) {
    asm volatile("cp.async.bulk.tensor.2d.global.shared::cta.tile.bulk_group [%0, {%1, %2}], [%3];" ::"l"(map), "r"(0),
                 "r"(row), "r"(skel::smem_addr(src))
                 : "memory");
}
__device__ __forceinline__ void tma_prefetch_desc(const skel_tmap *map) {
    asm volatile("prefetch.tensormap [%0];" ::"l"(map) : "memory");
}
// issue the two 256-row boxes of tile `tile` into stage buffer `dst`
template <int ROWS = RB>
__device__ __forceinline__ void issue_tile(unsigned char *dst, const skel_tmap *map, skel_u64 tile, skel_u64 *bar) {
    constexpr unsigned BYTES = (unsigned)ROWS * 128u;
    skel::mbar_expect_tx(bar, BYTES);
    const int row = (int)(tile * ROWS);
    tma_load_rows(dst, map, row, bar);
    tma_load_rows(dst + BYTES / 2, map, row + ROWS / 2, bar);
}
// thread `r` reads its 128-byte row of a 128B-swizzled stage into x[K]
// (templates so that element sizes without a TMA path never instantiate them)
template <bool OK = TMA_OK> __device__ __forceinline__ void read_row(const unsigned char *stage, int r, skel_T *x) {
    if constexpr (OK) {
        constexpr int PER = OK ? (int)(16 / sizeof(skel_T)) : 1;  // dependent: no arr<T,0> when !OK
        const unsigned char *row = stage + (size_t)r * 128;
#pragma unroll
        for (int j = 0; j < 8; ++j) {
            const uint4 q = *reinterpret_cast<const uint4 *>(row + ((j ^ (r & 7)) << 4));
            const auto e = skel::bit_cast<skel::arr<skel_T, PER>>(q);
#pragma unroll
            for (int k = 0; k < PER; ++k) x[j * PER + k] = e.v[k];
        }
    }
}
template <bool OK = TMA_OK> __device__ __forceinline__ void write_row(unsigned char *stage, int r, const skel_T *x) {
    if constexpr (OK) {
        constexpr int PER = OK ? (int)(16 / sizeof(skel_T)) : 1;  // dependent: no arr<T,0> when !OK
        unsigned char *row = stage + (size_t)r * 128;
#pragma unroll
        for (int j = 0; j < 8; ++j) {
            skel::arr<skel_T, PER> e;
#pragma unroll
            for (int k = 0; k < PER; ++k) e.v[k] = x[j * PER + k];
            *reinterpret_cast<uint4 *>(row + ((j ^ (r & 7)) << 4)) = skel::bit_cast<uint4>(e);
        }
    }
}
__device__ __forceinline__ unsigned char *aligned_stages(unsigned char *p) {
    const unsigned a = skel::smem_addr(p);
    return p + ((1024u - (a & 1023u)) & 1023u);
}

extern __shared__ __align__(16) unsigned char skel_dsmem[];

// ============================================================================
// Reduce
// ============================================================================
#ifndef SKEL_RED_MINB
#if SKEL_RED_DIRECT
#define SKEL_RED_MINB 4
#else
#define SKEL_RED_MINB 1
#endif
#endif
// a / b in 32-bit arithmetic when both fit (the 64-bit division is a
// subroutine call of ~100 instructions ahead of the first load)
__device__ __forceinline__ skel_u64 udiv(skel_u64 a, skel_u64 b) {
    if (((a | b) >> 32) == 0) return (unsigned)a / (unsigned)b;
    return a / b;
}
// ordered warp fold of 32 valid values: lane 0 receives x_0 (+) ... (+) x_31
template <class Tup> __device__ __forceinline__ skel_T warp_fold_full(skel_T x, int lane, Tup &t) {
#pragma unroll
    for (int d = 1; d < 32; d <<= 1) {
        const skel_T o = skel::shfl_down(x, d);
        if ((lane & (2 * d - 1)) == 0) x = opf(x, o, t);
    }
    return x;
}
__device__ __forceinline__ uint4 ld_stream16(const void *p) {
    uint4 q;
    asm volatile("ld.global.nc.L1::no_allocate.v4.u32 {%0,%1,%2,%3}, [%4];"
                 : "=r"(q.x), "=r"(q.y), "=r"(q.z), "=r"(q.w)
                 : "l"(p));
    return q;
}
// in-order fold of the PERV elements of one 16-byte lane load
template <bool OK = TMA_OK, class Tup> __device__ __forceinline__ skel_T fold16(const uint4 &q, Tup &t) {
    if constexpr (OK) {
        const auto e = skel::bit_cast<skel::arr<skel_T, PERV>>(q);
        skel_T a = e.v[0];
#pragma unroll
        for (int k = 1; k < PERV; ++k) a = opf(a, e.v[k], t);
        return a;
    } else {
        return skel_T{};
    }
}
__device__ __forceinline__ VT vt_make(const skel_T &v) {
    VT r;
    r.v = v;
    r.ok = true;
    return r;
}
// Direct Reduce of this CTA's range, valid in thread 0 (RDIRECT).  The n
// elements form warp-chunks of 32 consecutive lane loads (16 bytes each when
// `vec`, else one element); the G*NW warps of the grid own contiguous chunk
// ranges, each folds its range in order (lane fold, ordered shuffle tree per
// chunk, running aggregate in lane 0) with RU loads in flight per lane; the
// ragged tail (< one chunk) goes to the last warp; the CTA folds its warps in
// order.  No barrier inside the loop.
template <class Tup>
__device__ __forceinline__ VT reduce_direct(const skel_T *__restrict__ in, skel_u64 n, bool vec, VT *wpart, Tup &tup) {
    const int t = threadIdx.x, lane = t & 31, w = t >> 5;
    const skel_u64 G = gridDim.x, c = blockIdx.x;
    const skel_u64 per_chunk = (TMA_OK && vec) ? 32ull * PERV : 32ull;
    const skel_u64 nch = n / per_chunk;
    const skel_u64 NWT = G * NW, gw = c * NW + w;
    const skel_u64 k0 = udiv(nch * gw, NWT), k1 = udiv(nch * (gw + 1), NWT);
    VT wrun;
    wrun.ok = false;
    skel_u64 k = k0;
    if (TMA_OK && vec) {
        const uint4 *base = reinterpret_cast<const uint4 *>(in) + lane;
        for (; k + RU <= k1; k += RU) {
            uint4 q[RU];
#pragma unroll
            for (int u = 0; u < RU; ++u) q[u] = ld_stream16(base + (k + u) * 32);
#pragma unroll
            for (int u = 0; u < RU; ++u) {
                const skel_T a = warp_fold_full(fold16(q[u], tup), lane, tup);
                if (lane == 0) wrun = comb(wrun, vt_make(a), tup);
            }
        }
        for (; k < k1; ++k) {
            const skel_T a = warp_fold_full(fold16(ld_stream16(base + k * 32), tup), lane, tup);
            if (lane == 0) wrun = comb(wrun, vt_make(a), tup);
        }
    } else {
        const skel_T *base = in + lane;
        for (; k + RU <= k1; k += RU) {
            skel_T q[RU];
#pragma unroll
            for (int u = 0; u < RU; ++u) q[u] = base[(k + u) * 32];
#pragma unroll
            for (int u = 0; u < RU; ++u) {
                const skel_T a = warp_fold_full(q[u], lane, tup);
                if (lane == 0) wrun = comb(wrun, vt_make(a), tup);
            }
        }
        for (; k < k1; ++k) {
            const skel_T a = warp_fold_full(base[k * 32], lane, tup);
            if (lane == 0) wrun = comb(wrun, vt_make(a), tup);
        }
    }
    if (gw == NWT - 1) {  // ragged tail, in order after the last chunk
        const skel_u64 b0 = nch * per_chunk, rem = n - b0;
        if (rem) {
            const skel_u64 kt = (rem + 31) / 32;
            VT a;
            a.ok = false;
            for (skel_u64 j2 = 0; j2 < kt; ++j2) {
                const skel_u64 j = (skel_u64)lane * kt + j2;
                if (j < rem) a = comb(a, vt_make(in[b0 + j]), tup);
            }
            a = warp_fold(a, lane, tup);
            if (lane == 0) wrun = comb(wrun, a, tup);
        }
    }
    if (lane == 0) wpart[w] = wrun;
    __syncthreads();
    VT r;
    r.ok = false;
    if (w == 0) {
        VT y;
        y.ok = false;
        if (lane < NW) y = wpart[lane];
        r = warp_fold(y, lane, tup);
    }
    return r;
}

// ---- cross-device single pass --
// A block-distributed Reduce over K in-process devices without a separate
// exchange: the one thread that ends a device's Reduce publishes the device's
// result into slot k of an array in logical device 0's memory (over NVLink
// for another GPU), then takes a ticket from a counter there (release/acquire
// at system scope).  The device that draws the last ticket folds the K
// published values IN DEVICE ORDER (eq. (3) with a non-commutative operator
// stays exact) and stores the result into every device's result slot, then
// resets the counter.  Nobody waits for anybody -- the last arriver does the
// fold -- so kernels of logical devices that share one GPU cannot deadlock.
// It also copies the K device results to every device (a block-distributed
// Scan seeds device k with results 0..k-1).  The host joins the devices' streams after the launches (every later use,
// and the next Reduce's tickets, come after the last arriver's stores).
#define SKEL_XMAX 16
struct skel_xdev {
    skel_S *slots;           // K published device results (logical device 0's memory)
    unsigned *ticket;        // arrivals (logical device 0's memory)
    skel_S *dst[SKEL_XMAX];  // result slot of every local device
    skel_S *gat[SKEL_XMAX];  // every local device's copy of the K device results (the
                             // cross-device Scan seeds device k from results 0..k-1)
    int k, K, ndst;          // this device, devices holding data, local devices
};
template <class Tup> __device__ __forceinline__ void skel_xdev_finish(const skel_xdev &xd, const skel_T &v, Tup &tup) {
    skel::st_value_sys(&xd.slots[xd.k], skel_S{v});
    skel::fence_acq_rel_sys();  // the value before the ticket
    const unsigned prev = skel::atom_add_acq_rel_sys(xd.ticket, 1u);
    if (prev != (unsigned)(xd.K - 1)) return;
    skel::fence_acq_rel_sys();  // every device's value after its ticket
    skel_T acc = skel::ld_value_sys(&xd.slots[0]).v;
    for (int j = 1; j < xd.K; ++j) acc = opf(acc, skel::ld_value_sys(&xd.slots[j]).v, tup);
    for (int d = 0; d < xd.ndst; ++d) {
        skel::st_value_sys(xd.dst[d], skel_S{acc});
        if (xd.gat[d] != xd.slots)
            for (int j = 0; j < xd.K; ++j) skel::st_value_sys(&xd.gat[d][j], skel::ld_value_sys(&xd.slots[j]));
    }
    skel::st_relaxed_sys_u32(xd.ticket, 0u);
}

extern "C" __global__ void __launch_bounds__(RB, SKEL_RED_MINB)
    skel_reduce_kernel(const __grid_constant__ skel_tmap tin, const skel_T *__restrict__ in, skel_u64 n, int use_tma,
                       skel_S *partials, unsigned *pvalid, unsigned *counter, skel_S *result,
                       const __grid_constant__ skel_xdev xd, const skel_Buf args) {
    skel::pdl_wait();  // launched as a programmatic dependent (prelude.cuh)
    skel::pdl_trigger();
    auto tup = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    __shared__ skel_u64 bars[STAGES];
    __shared__ VT wpart[NW];
    __shared__ int s_last;
    const int t = threadIdx.x;
    const skel_u64 nft = n / TILE;
    const skel_u64 G = gridDim.x, c = blockIdx.x;
    const skel_u64 t0 = udiv(nft * c, G), t1 = udiv(nft * (c + 1), G);
    const skel_u64 my = RIL ? (nft > c ? (nft - c + G - 1) / G : 0) : t1 - t0;
    auto tile_at = [&](skel_u64 i) -> skel_u64 { return RIL ? c + i * G : t0 + i; };
    VT run;
    run.ok = false;
    // RIL: every tile's fold is a partial of its own (index = tile)
    auto take = [&](VT tv, skel_u64 tile) {
        if (RIL) {
            skel::st_value(&partials[tile], skel_S{tv.v});
        } else {
            run = comb(run, tv, tup);
        }
    };

    if (RDIRECT) {
        run = reduce_direct(in, n, use_tma != 0, wpart, tup);
    } else if (TMA_OK && use_tma) {
        unsigned char *stages = aligned_stages(skel_dsmem);
        if (t == 0) {
            for (int s = 0; s < STAGES; ++s) skel::mbar_init(&bars[s], 1);
            skel::fence_mbar_init();
            tma_prefetch_desc(&tin);
        }
        __syncthreads();
        if (t == 0)
            for (skel_u64 s = 0; s < STAGES && s < my; ++s) issue_tile(stages + s * TILE_BYTES, &tin, tile_at(s), &bars[s]);
        for (skel_u64 i = 0; i < my; ++i) {
            const int s = (int)(i % STAGES);
            skel::mbar_wait(&bars[s], (unsigned)((i / STAGES) & 1));
            skel_T x[K];
            read_row(stages + s * TILE_BYTES, t, x);
            VT a;
            a.v = x[0];
            a.ok = true;
#pragma unroll
            for (int k = 1; k < K; ++k) a.v = opf(a.v, x[k], tup);
            __syncthreads();  // stage s fully consumed
            if (t == 0 && i + STAGES < my) issue_tile(stages + s * TILE_BYTES, &tin, tile_at(i + STAGES), &bars[s]);
            VT tv = block_fold(a, wpart, tup);
            if (t == 0) take(tv, tile_at(i));
        }
    } else {
        for (skel_u64 i = 0; i < my; ++i) {
            const skel_T *p = in + tile_at(i) * TILE + (skel_u64)t * K;
            VT a;
            a.v = p[0];
            a.ok = true;
#pragma unroll 4
            for (int k = 1; k < K; ++k) a.v = opf(a.v, p[k], tup);
            __syncthreads();
            VT tv = block_fold(a, wpart, tup);
            if (t == 0) take(tv, tile_at(i));
        }
    }
    // ragged last tile: direct loads, owned by the last CTA (keeps index order)
    if (!RDIRECT && c == G - 1 && nft * TILE < n) {
        const skel_u64 base = nft * TILE, rem = n - base;
        const skel_u64 kt = (rem + RB - 1) / RB;
        VT a;
        a.ok = false;
        for (skel_u64 k = 0; k < kt; ++k) {
            const skel_u64 j = (skel_u64)t * kt + k;
            if (j < rem) {
                VT e;
                e.v = in[base + j];
                e.ok = true;
                a = comb(a, e, tup);
            }
        }
        __syncthreads();
        VT tv = block_fold(a, wpart, tup);
        if (t == 0) take(tv, nft);
    }
    // publish this CTA's partial (RIL: the tile partials are already out); the
    // last CTA to finish folds them in order
    const skel_u64 NP = (RIL && !RDIRECT) ? nft + (nft * TILE < n ? 1 : 0) : G;  // partials
    if (t == 0) {
        if (!RIL || RDIRECT) {
            skel::st_value(&partials[c], skel_S{run.v});
            skel::st_relaxed_u32(&pvalid[c], run.ok ? 1u : 0u);
        }
        // message passing through the counter: release fence before the
        // increment, acquire fence in the CTA that sees the last count (an
        // acq_rel fence, not the sequentially consistent __threadfence); the
        // barrier then orders the other threads' loads after it
        skel::fence_acq_rel_gpu();
        const unsigned prev = atomicAdd(counter, 1u);
        const bool last = prev == (unsigned)(G - 1);
        if (last) skel::fence_acq_rel_gpu();
        s_last = last;
    }
    __syncthreads();
    if (s_last) {
        const skel_u64 per = (NP + RB - 1) / RB;
        VT a;
        a.ok = false;
        // loads in batches of 8 (independent L2 round trips), folded in order
        for (skel_u64 k0 = 0; k0 < per; k0 += 8) {
            VT e[8];
#pragma unroll
            for (int u = 0; u < 8; ++u) {
                const skel_u64 j = (skel_u64)t * per + k0 + u;
                e[u].ok = k0 + u < per && j < NP && ((RIL && !RDIRECT) || skel::ld_relaxed_u32(&pvalid[j]));
                if (e[u].ok) e[u].v = skel::ld_value(&partials[j]).v;
            }
#pragma unroll
            for (int u = 0; u < 8; ++u) a = comb(a, e[u], tup);
        }
        VT r = block_fold(a, wpart, tup);
        if (t == 0) {
            result->v = r.v;
            *counter = 0;
            if (xd.K) skel_xdev_finish(xd, r.v, tup);
        }
    }
}

// fold count >= 1 published values in order (cross-device Reduce)
extern "C" __global__ void skel_fold_kernel(const skel_S *vals, int count, skel_S *out, const skel_Buf args) {
    skel::pdl_wait();
    skel::pdl_trigger();
    auto tup = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    if (threadIdx.x == 0 && blockIdx.x == 0) {
        skel_T acc = vals[0].v;
        for (int i = 1; i < count; ++i) acc = opf(acc, vals[i].v, tup);
        out->v = acc;
    }
}
// seed of logical device k in a block-distributed Scan: id for k == 0,
// otherwise agg_0 (+) ... (+) agg_{k-1}
extern "C" __global__ void skel_seed_kernel(const skel_S *aggs, int k, const skel_S identity, skel_S *out,
                                            const skel_Buf args) {
    skel::pdl_wait();
    skel::pdl_trigger();
    auto tup = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    if (threadIdx.x == 0 && blockIdx.x == 0) {
        if (k == 0) {
            out->v = identity.v;
        } else {
            skel_T acc = aggs[0].v;
            for (int i = 1; i < k; ++i) acc = opf(acc, aggs[i].v, tup);
            out->v = acc;
        }
    }
}

// ============================================================================
// Scan: single pass over HBM with an L2-resident second read
//
// A persistent grid of G CTAs (one per SM) walks the vector in *slices* of
// G x CH tiles; CTA c owns the CH consecutive tiles (s*G + c)*CH ... of slice
// s.  Per slice and CTA:
//   P1(s): fold the CTA's tiles in order (TMA loads with an L2 evict_last
//          policy, so the slice stays in L2) and publish the aggregate A(s,c);
//   P2(s): prefix(s,c) = carry(s) (+) A(s,0) (+) ... (+) A(s,c-1), with
//          carry(s) = carry(s-1) (+) A(s-1,0) (+) ... (+) A(s-1,G-1); then
//          re-read the tiles (L2 hits, evict_first), scan them with a running
//          prefix and TMA-store the outputs (evict_first).
// Work order per CTA: P1(0), P1(1), P2(0), P1(2), P2(1), ... so each CTA's
// wait for its predecessors' aggregates of slice s is covered by its own
// P1(s+1): no CTA waits on another in the steady state, HBM sees each input
// byte read once and each output byte written once (8 B/element for float),
// and every element's prefix chain has one carry link per slice (float
// rounding stays far below 1e-5 at 2^30 elements).
// The ragged last tile is scanned by CTA G-1 with direct loads; element sizes
// without a TMA path use direct loads for every tile.
// ============================================================================
#ifndef SKEL_SCAN_KEEP_POLICY
#define SKEL_SCAN_KEEP_POLICY evict_last
#endif
#ifndef SKEL_SCAN_DROP_POLICY
#define SKEL_SCAN_DROP_POLICY evict_first
#endif
#define SKEL_STR2(x) #x
#define SKEL_STR(x) SKEL_STR2(x)
// L2 policy of the P1 loads (the slice must survive until P2 re-reads it)
__device__ __forceinline__ skel_u64 policy_evict_last() {
    skel_u64 p;
    asm volatile("createpolicy.fractional.L2::" SKEL_STR(SKEL_SCAN_KEEP_POLICY) ".b64 %0, 1.0;" : "=l"(p));
    return p;
}
// L2 policy of the P2 loads and of the output stores (dead after use)
__device__ __forceinline__ skel_u64 policy_evict_first() {
    skel_u64 p;
    asm volatile("createpolicy.fractional.L2::" SKEL_STR(SKEL_SCAN_DROP_POLICY) ".b64 %0, 1.0;" : "=l"(p));
    return p;
}
__device__ __forceinline__ void tma_load_rows_hint(void *dst, const skel_tmap *map, int row, skel_u64 *bar,
                                                   skel_u64 pol) {
    asm volatile(
        "cp.async.bulk.tensor.2d.shared::cluster.global.tile.mbarrier::complete_tx::bytes.L2::cache_hint"
        " [%0], [%1, {%2, %3}], [%4], %5;" ::"r"(skel::smem_addr(dst)),
        "l"(map), "r"(0), "r"(row), "r"(skel::smem_addr(bar)), "l"(pol)
        : "memory");
}
__device__ __forceinline__ void tma_store_rows_hint(const skel_tmap *map, int row, const void *src, skel_u64 pol) {
    asm volatile("cp.async.bulk.tensor.2d.global.shared::cta.tile.bulk_group.L2::cache_hint [%0, {%1, %2}], [%3], %4;" ::"l"(
                     map),
                 "r"(0), "r"(row), "r"(skel::smem_addr(src)), "l"(pol)
                 : "memory");
}

// status of A(s,c): state 1 = value, 2 = empty sub-chunk
__device__ __forceinline__ void publish_agg(skel_u64 *st64, unsigned *fl32, skel_S *vals, skel_u64 idx, unsigned epoch,
                                            const VT &a) {
    const unsigned state = a.ok ? 1u : 2u;
    if constexpr (PACKED) {
        skel_S sv{a.v};
        const unsigned bits = skel::bit_cast<unsigned>(sv);
        const skel_u64 word = ((skel_u64)bits << 32) | (skel_u64)((epoch << 2) | state);
        // value, epoch and state travel in ONE 64-bit word, so nothing else has
        // to be ordered before it: a relaxed store suffices (a release would
        // cost a GPU-scope fence -- microseconds under streaming load -- on the
        // consumers' critical path)
        asm volatile("st.relaxed.gpu.global.u64 [%0], %1;" ::"l"(st64 + idx), "l"(word) : "memory");
    } else {
        if (a.ok) skel::st_value(&vals[idx], skel_S{a.v});
        skel::st_release(&fl32[idx], (epoch << 2) | state);
    }
}
// spin until A(idx) is published; returns it
__device__ __forceinline__ VT wait_agg(const skel_u64 *st64, const unsigned *fl32, const skel_S *vals, skel_u64 idx,
                                       unsigned epoch) {
    VT r;
    if constexpr (PACKED) {
        skel_u64 word;
        do {
            asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(word) : "l"(st64 + idx) : "memory");
        } while (((unsigned)word >> 2) != epoch);
        r.ok = ((unsigned)word & 3u) == 1u;
        r.v = skel::bit_cast<skel_S>((unsigned)(word >> 32)).v;
    } else {
        unsigned f;
        do {
            f = skel::ld_acquire(&fl32[idx]);
        } while ((f >> 2) != epoch);
        r.ok = (f & 3u) == 1u;
        if (r.ok) r.v = skel::ld_value(&vals[idx]).v;
    }
    return r;
}
// relaxed probe of A(idx): true once published in this epoch
__device__ __forceinline__ bool probe_agg(const skel_u64 *st64, const unsigned *fl32, const skel_S *vals, skel_u64 idx,
                                          unsigned epoch, VT &r) {
    if constexpr (PACKED) {
        skel_u64 word;
        asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(word) : "l"(st64 + idx) : "memory");
        if (((unsigned)word >> 2) != epoch) return false;
        r.ok = ((unsigned)word & 3u) == 1u;
        r.v = skel::bit_cast<skel_S>((unsigned)(word >> 32)).v;
        return true;
    } else {
        const unsigned f = skel::ld_acquire(&fl32[idx]);
        if ((f >> 2) != epoch) return false;
        r.ok = (f & 3u) == 1u;
        if (r.ok) r.v = skel::ld_value(&vals[idx]).v;
        return true;
    }
}
constexpr int AGG_PER = 16;  // status words one prefix-warp lane polls at most
#ifndef SKEL_SCAN_NPRE
#define SKEL_SCAN_NPRE 4
#endif
constexpr int NPRE = SKEL_SCAN_NPRE;  // slice windows buffered for the consumers
#ifndef SKEL_SCAN_BACKOFF_MIN
#define SKEL_SCAN_BACKOFF_MIN 32
#endif
#ifndef SKEL_SCAN_BACKOFF_MAX
#define SKEL_SCAN_BACKOFF_MAX 1024
#endif

// ordered fold of A(base .. base+cnt-1) by one warp (cnt <= 32*AGG_PER);
// every lane issues all of its probes before waiting; result in every lane
template <class Tup>
__device__ __forceinline__ VT warp_fold_aggs(const skel_u64 *st64, const unsigned *fl32, const skel_S *vals,
                                             skel_u64 base, int cnt, unsigned epoch, int lane, Tup &t) {
    const int per = (cnt + 31) / 32;
    VT e[AGG_PER];
    bool got[AGG_PER];
#pragma unroll
    for (int k = 0; k < AGG_PER; ++k) got[k] = !(k < per && lane * per + k < cnt);
    for (unsigned ns = SKEL_SCAN_BACKOFF_MIN;; ns = ns < SKEL_SCAN_BACKOFF_MAX ? 2 * ns : ns) {
        bool all = true;
#pragma unroll
        for (int k = 0; k < AGG_PER; ++k) {
            if (!got[k]) {
                got[k] = probe_agg(st64, fl32, vals, base + lane * per + k, epoch, e[k]);
                all = all && got[k];
            }
        }
        if (__all_sync(0xffffffffu, all)) break;
        __nanosleep(ns);  // back off: many CTAs poll the same status lines
    }
    VT a;
    a.ok = false;
#pragma unroll
    for (int k = 0; k < AGG_PER; ++k)
        if (k < per && lane * per + k < cnt) a = comb(a, e[k], t);
    a = warp_fold(a, lane, t);
    return vt_shfl_idx(a, 0);
}

#ifndef SKEL_SCAN_CPOLL
#define SKEL_SCAN_CPOLL 1
#endif
// the same ordered fold with coalesced probes (packed status words only): probe
// round k reads words base + 32k + lane, so one round touches 2 L2 lines instead
// of `per` rounds each spanning 32 lines (4x fewer sector requests per poll on
// the hot status lines); the words are transposed through shared memory so each
// lane folds `per` consecutive aggregates in order before the warp fold
template <class Tup>
__device__ __forceinline__ VT warp_fold_aggs_coalesced(const skel_u64 *st64, skel_u64 *sbuf, skel_u64 base, int cnt,
                                                       unsigned epoch, int lane, Tup &t) {
    const int rounds = (cnt + 31) / 32;
    unsigned pending = 0;  // bit k: word base + 32k + lane still unpublished
#pragma unroll
    for (int k = 0; k < AGG_PER; ++k)
        if (k < rounds && 32 * k + lane < cnt) pending |= 1u << k;
    for (unsigned ns = SKEL_SCAN_BACKOFF_MIN;; ns = ns < SKEL_SCAN_BACKOFF_MAX ? 2 * ns : ns) {
        skel_u64 word[AGG_PER];
#pragma unroll
        for (int k = 0; k < AGG_PER; ++k)
            if (pending >> k & 1u)
                asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];"
                             : "=l"(word[k])
                             : "l"(st64 + base + 32 * k + lane)
                             : "memory");
#pragma unroll
        for (int k = 0; k < AGG_PER; ++k)
            if ((pending >> k & 1u) && ((unsigned)word[k] >> 2) == epoch) {
                sbuf[32 * k + lane] = word[k];
                pending &= ~(1u << k);
            }
        if (__all_sync(0xffffffffu, pending == 0)) break;
        __nanosleep(ns);
    }
    __syncwarp();
    const int per = (cnt + 31) / 32;
    VT a;
    a.ok = false;
#pragma unroll
    for (int k = 0; k < AGG_PER; ++k) {
        const int i = lane * per + k;
        if (k < per && i < cnt) {
            const skel_u64 w = sbuf[i];
            VT x;
            x.ok = ((unsigned)w & 3u) == 1u;
            x.v = skel::bit_cast<skel_S>((unsigned)(w >> 32)).v;
            a = comb(a, x, t);
        }
    }
    __syncwarp();  // sbuf is reused by the next window
    a = warp_fold(a, lane, t);
    return vt_shfl_idx(a, 0);
}


// work item q of a CTA's sequence: P1 of slices 0..LAG-1, then per slice s:
// P1(s+LAG) x CH (if that slice exists), P2(s) x CH.  Returns false past the
// end.  LAG slices of slack absorb the CTAs' speed differences.
#ifndef SKEL_SCAN_LAG
#define SKEL_SCAN_LAG 2
#endif
constexpr int SCAN_LAG = SKEL_SCAN_LAG;
__device__ __forceinline__ bool scan_item(skel_u64 q, skel_u64 nslices, int &phase, skel_u64 &s, int &j) {
    const skel_u64 L = SCAN_CH;
    const skel_u64 P = nslices < (skel_u64)SCAN_LAG ? nslices : (skel_u64)SCAN_LAG;
    if (q < P * L) {
        phase = 1;
        s = q / L;
        j = (int)(q % L);
        return true;
    }
    const skel_u64 k = q - P * L;
    const skel_u64 F = nslices > (skel_u64)SCAN_LAG ? nslices - SCAN_LAG : 0;
    if (k < F * 2 * L) {
        const skel_u64 blk = k / (2 * L), r = k % (2 * L);
        phase = r < L ? 1 : 2;
        s = r < L ? blk + SCAN_LAG : blk;
        j = (int)(r < L ? r : r - L);
        return true;
    }
    const skel_u64 k2 = k - F * 2 * L;
    s = F + k2 / L;
    if (s >= nslices) return false;
    phase = 2;
    j = (int)(k2 % L);
    return true;
}

#ifdef SKEL_SCAN_TRACE
// lab instrumentation (tools/scan_lab.cu): globaltimer stamps per (slice, CTA)
//   0 = P1 aggregate published, 1 = prefix ready, 2 = P2 start, 3 = P2 done,
//   4 = prefix warp starts the slice
__device__ skel_u64 skel_scan_trace[6 * 148 * 1024];
__device__ __forceinline__ void scan_stamp(int ev, skel_u64 s, skel_u64 c) {
    skel_u64 t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    if (s < 1024 && c < 148) skel_scan_trace[(ev * 1024 + s) * 148 + c] = t;
}
#define SKEL_STAMP(ev, s, c) scan_stamp(ev, s, c)
#else
#define SKEL_STAMP(ev, s, c)
#endif
// consumers = the SRB threads of warps 0..SNW-1; warp SNW is the TMA producer,
// warp SNW+1 issues the TMA stores of scanned tiles and hands their stages back,
// warps SNW+2 .. SNW+1+PW fold the slice windows ahead of the consumers
constexpr int SCAN_THREADS = SRB + 64 + 32 * PW;
__device__ __forceinline__ void cons_sync() { asm volatile("bar.sync 1, %0;" ::"n"(SRB) : "memory"); }
__device__ __forceinline__ void mbar_arrive(skel_u64 *bar) {
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(skel::smem_addr(bar)) : "memory");
}
// ordered fold over the consumers; result in thread 0
template <class Tup> __device__ __forceinline__ VT cons_fold(VT x, VT *wpart, Tup &t) {
    const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
    x = warp_fold(x, lane, t);
    if (lane == 0) wpart[w] = x;
    cons_sync();
    VT r;
    r.ok = false;
    if (w == 0) {
        VT y;
        y.ok = false;
        if (lane < SNW) y = wpart[lane];
        r = warp_fold(y, lane, t);
    }
    return r;
}
// ordered exclusive scan over the consumers with ONE barrier: warp totals go
// to wbuf, then every warp scans the SNW totals itself (redundantly) to get
// its warp prefix and the block total.  Callers alternate two wbuf buffers
// between consecutive tiles, so a buffer is rewritten only after a barrier
// that every reader of its previous contents has passed.
template <class Tup> __device__ __forceinline__ VT cons_exscan1(VT x, VT *wbuf, VT &total, Tup &t) {
    const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
    VT inc = x;
#pragma unroll
    for (int d = 1; d < 32; d <<= 1) {
        VT o = vt_shfl_up(inc, d);
        if (lane >= d) inc = comb(o, inc, t);
    }
    VT ex = vt_shfl_up(inc, 1);
    if (lane == 0) ex.ok = false;
    if (lane == 31) wbuf[w] = inc;
    cons_sync();
    VT yi;
    yi.ok = false;
    if (lane < SNW) yi = wbuf[lane];
#pragma unroll
    for (int d = 1; d < SNW; d <<= 1) {
        VT o = vt_shfl_up(yi, d);
        if (lane >= d) yi = comb(o, yi, t);
    }
    VT wpre = vt_shfl_idx(yi, w > 0 ? w - 1 : 0);
    if (w == 0) wpre.ok = false;
    total = vt_shfl_idx(yi, SNW - 1);
    return comb(wpre, ex, t);
}

#ifndef SKEL_SCAN_MINB
#define SKEL_SCAN_MINB 1
#endif
extern "C" __global__ void __launch_bounds__(SCAN_THREADS, SKEL_SCAN_MINB)
    skel_scan_kernel(const __grid_constant__ skel_tmap tin, const __grid_constant__ skel_tmap tout,
                     const skel_T *in, skel_T *out, skel_u64 n, int use_tma, const skel_S identity, const skel_S *seed,
                     skel_u64 *status, unsigned *flags, skel_S *aggv, skel_S *incv, unsigned *counters,
                     unsigned *epoch_ptr, skel_S *total, const skel_Buf args) {
    (void)incv;
    // launched cooperatively AND as a programmatic dependent of the previous
    // kernel: nothing is touched (and no CTA waits on another) before that
    // kernel has completed, by which time the whole grid is resident
    skel::pdl_wait();
    skel::pdl_trigger();
    // the launch's epoch lives in device memory (graph replays must see a new
    // one): every CTA reads it before publishing anything; the last CTA to
    // finish advances it (all CTAs have read it by then)
    auto tup = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    __shared__ unsigned s_epoch;
    // full: TMA load landed; empty: stage free (P1: consumers done reading,
    // P2: the store of its outputs has read it); outs: P2 outputs staged
    __shared__ skel_u64 full_bar[SSTAGES], empty_bar[SSTAGES], outs_bar[SSTAGES], pre_full[NPRE], pre_empty[NPRE];
    __shared__ VT wsc[2][SNW];  // warp partials, alternated between consecutive tiles
    __shared__ VT s_pre[NPRE];
    __shared__ skel_u64 s_win[(PACKED && SKEL_SCAN_CPOLL) ? PW * 32 * AGG_PER : 1];  // coalesced-poll transpose
    const int t = threadIdx.x, lane = t & 31, w = t >> 5;
    const skel_u64 G = gridDim.x, c = blockIdx.x;
    const skel_u64 nft = n / STILE;  // full tiles
    const skel_u64 per_slice = G * SCAN_CH;
    const skel_u64 nslices = udiv(nft + per_slice - 1, per_slice);
    const skel_u64 rstride = (nslices * G + 63) / 64 * 64;  // status words per copy
    const bool tma = TMA_OK && use_tma;
    unsigned char *stages = aligned_stages(skel_dsmem);
    auto tile_of = [&](skel_u64 s, int j) -> skel_u64 { return (s * G + c) * SCAN_CH + (skel_u64)j; };
    auto jn = [&](skel_u64 s) -> int {  // valid tiles of this CTA in slice s
        const skel_u64 first = (s * G + c) * SCAN_CH;
        if (first >= nft) return 0;
        const skel_u64 left = nft - first;
        return (int)(left < (skel_u64)SCAN_CH ? left : (skel_u64)SCAN_CH);
    };
    // a window folds G-1 aggregates with one warp (<= 32 x AGG_PER); the host
    // caps the grid at 513 CTAs -- a larger grid would fold silently wrong
    if (G - 1 > (skel_u64)(32 * AGG_PER)) __trap();
    if (t == 0) {
        for (int st = 0; st < SSTAGES; ++st) {
            skel::mbar_init(&full_bar[st], 1);
            skel::mbar_init(&empty_bar[st], 1);
            skel::mbar_init(&outs_bar[st], SRB);
        }
        for (int k = 0; k < NPRE; ++k) {
            skel::mbar_init(&pre_full[k], 1);
            skel::mbar_init(&pre_empty[k], SRB);
        }
        skel::fence_mbar_init();
        s_epoch = *(volatile unsigned *)epoch_ptr;
    }
    __syncthreads();
    const unsigned epoch = s_epoch;

    if (w == SNW) {
        // ================================================ TMA producer warp
        if (tma && lane == 0) {
            const skel_u64 pol_keep = policy_evict_last(), pol_drop = policy_evict_first();
            tma_prefetch_desc(&tin);
            skel_u64 v = 0;
            int ph, j;
            skel_u64 s;
            for (skel_u64 q = 0; scan_item(q, nslices, ph, s, j); ++q) {
                if (j >= jn(s)) continue;
                const int st = (int)(v % SSTAGES);
                if (v >= SSTAGES) skel::mbar_wait(&empty_bar[st], (unsigned)((v / SSTAGES - 1) & 1));
                const int row = (int)(tile_of(s, j) * SRB);
                unsigned char *dst = stages + st * STILE_BYTES;
                const skel_u64 pol = ph == 1 ? pol_keep : pol_drop;
                skel::mbar_expect_tx(&full_bar[st], STILE_BYTES);
                tma_load_rows_hint(dst, &tin, row, &full_bar[st], pol);
                tma_load_rows_hint(dst + STILE_BYTES / 2, &tin, row + SRB / 2, &full_bar[st], pol);
                ++v;
            }
        }
        return;
    }

    if (w == SNW + 1) {
        // ================================================ TMA store warp
        // stores each scanned tile as soon as its outputs are staged; the
        // stage goes back to the producer once the store has read it
        if (tma && lane == 0) {
            const skel_u64 pol_drop = policy_evict_first();
            tma_prefetch_desc(&tout);
            skel_u64 v = 0;
            unsigned par = 0;  // phase parity of outs_bar[st], one bit per stage
            int ph, j;
            skel_u64 s;
            for (skel_u64 q = 0; scan_item(q, nslices, ph, s, j); ++q) {
                if (j >= jn(s)) continue;
                const int st = (int)(v % SSTAGES);
                ++v;
                if (ph != 2) continue;
                skel::mbar_wait(&outs_bar[st], (par >> st) & 1u);
                par ^= 1u << st;
                const int row = (int)(tile_of(s, j) * SRB);
                unsigned char *src = stages + st * STILE_BYTES;
                tma_store_rows_hint(&tout, row, src, pol_drop);
                tma_store_rows_hint(&tout, row + SRB / 2, src + STILE_BYTES / 2, pol_drop);
                skel::bulk_commit();
                skel::bulk_wait_read0();
                mbar_arrive(&empty_bar[st]);
            }
            skel::bulk_wait0();
        }
        return;
    }

    if (w >= SNW + 2) {
        // ================================================ window warps
        // The consumers carry the running prefix from slice to slice: after P2(s-1)
        // their prefix is p(s-1) (+) A(s-1,c), so
        //   p(s) = that (+) A(s-1,c+1..G-1) (+) A(s,0..c-1)  =: that (+) W(s),
        // a window of G-1 consecutive aggregates (W(0) = A(0,0..c-1)).  Windows of
        // different slices are independent, so PW warps fold them concurrently
        // (warp k takes s = k, k+PW, ...): an L2 poll takes microseconds while the
        // SM streams, and one warp folding one window per round trip would pace
        // the whole grid.  Results go to a ring of NPRE slots the consumers drain.
        const int k = w - (SNW + 2);
        for (skel_u64 s = (skel_u64)k; s < nslices; s += PW) {
            const int slot = (int)(s % NPRE);
            if (s >= (skel_u64)NPRE) skel::mbar_wait(&pre_empty[slot], (unsigned)((s / NPRE - 1) & 1));
            if (lane == 0) SKEL_STAMP(4, s, c);
            const skel_u64 base = s == 0 ? 0 : (s - 1) * G + c + 1;
            const int cnt = s == 0 ? (int)c : (int)G - 1;
            VT win;
            win.ok = false;
            if (cnt > 0) {
                if constexpr (PACKED && SKEL_SCAN_CPOLL)
                    win = warp_fold_aggs_coalesced(status + (c % REPL) * rstride, s_win + k * 32 * AGG_PER, base, cnt,
                                                   epoch, lane, tup);
                else
                    win = warp_fold_aggs(status + (c % REPL) * rstride, flags, aggv, base, cnt, epoch, lane, tup);
            }
            if (lane == 0) {
                SKEL_STAMP(1, s, c);
                s_pre[slot] = win;
                mbar_arrive(&pre_full[slot]);
            }
            __syncwarp();
        }
        return;
    }

    // ==================================================== consumer warps
    skel_u64 v = 0;  // valid items consumed
    VT run1;         // P1 running aggregate of this CTA's sub-chunk (thread 0)
    run1.ok = false;
    VT run;          // P2 running prefix (identical in every consumer thread)
    run.v = seed ? seed->v : identity.v;
    run.ok = true;
    int ph, j;
    skel_u64 s;
    for (skel_u64 q = 0; scan_item(q, nslices, ph, s, j); ++q) {
        const int nj = jn(s);
        if (ph == 2 && j == 0) {  // p(s) = p(s-1) (+) own A(s-1,c) (+) W(s), W folded ahead
            const int slot = (int)(s % NPRE);
            skel::mbar_wait(&pre_full[slot], (unsigned)((s / NPRE) & 1));
            run = comb(run, s_pre[slot], tup);
            mbar_arrive(&pre_empty[slot]);
            if (t == 0) SKEL_STAMP(2, s, c);
        }
        if (j >= nj) {
            if (ph == 1 && j == 0 && nj == 0 && t == 0) {  // empty sub-chunk: publish once
                VT e;
                e.ok = false;
                for (int r = 0; r < REPL; ++r) publish_agg(status + r * rstride, flags, aggv, s * G + c, epoch, e);
            }
            continue;
        }
        const int st = (int)(v % SSTAGES);
        const skel_u64 tile = tile_of(s, j);
        skel_T x[K];
        if (tma) {
            skel::mbar_wait(&full_bar[st], (unsigned)((v / SSTAGES) & 1));
            read_row(stages + st * STILE_BYTES, t, x);
        } else {
            const skel_T *p = in + tile * STILE + (skel_u64)t * K;
#pragma unroll
            for (int k = 0; k < K; ++k) x[k] = p[k];
        }
        if (ph == 1) {
            // ---- P1: ordered fold of the tile
            VT a;
            a.v = x[0];
            a.ok = true;
#pragma unroll
            for (int k = 1; k < K; ++k) a.v = opf(a.v, x[k], tup);
            const VT tv = cons_fold(a, wsc[v & 1], tup);  // its barrier: every row is read
            if (t == 0) {
                if (tma) mbar_arrive(&empty_bar[st]);  // stage free for the producer
                run1 = comb(run1, tv, tup);
                if (j == nj - 1) {
                    SKEL_STAMP(0, s, c);
                    for (int r = 0; r < REPL; ++r)
                        publish_agg(status + r * rstride, flags, aggv, s * G + c, epoch, run1);
                    run1.ok = false;
                }
            }
        } else {
            // ---- P2: scan of the tile with the running prefix
#pragma unroll
            for (int k = 1; k < K; ++k) x[k] = opf(x[k - 1], x[k], tup);
            VT mine;
            mine.v = x[K - 1];
            mine.ok = true;
            VT tot;
            const VT excl = cons_exscan1(mine, wsc[v & 1], tot, tup);
            const VT pre = comb(run, excl, tup);
            run = comb(run, tot, tup);
#pragma unroll
            for (int k = K - 1; k >= 1; --k) x[k] = opf(pre.v, x[k - 1], tup);
            x[0] = pre.v;
            if (tma) {
                write_row(stages + st * STILE_BYTES, t, x);
                skel::fence_proxy_async();
                mbar_arrive(&outs_bar[st]);  // outputs staged: the store warp writes them
                if (t == 0 && j == nj - 1) SKEL_STAMP(3, s, c);
            } else {
                skel_T *o = out + tile * STILE + (skel_u64)t * K;
#pragma unroll
                for (int k = 0; k < K; ++k) o[k] = x[k];
            }
        }
        ++v;
    }
    // ---- ragged last tile and the device total: CTA G-1
    if (c == G - 1) {
        const VT carry_end = run;  // p(nslices): CTA G-1 has no later aggregates in its window
        const skel_u64 base = nft * STILE;
        VT mine;
        mine.ok = false;
        skel_u64 first = 0, kt = 0;
        if (base < n) {
            const skel_u64 cnt = n - base, per = (cnt + SRB - 1) / SRB;
            first = base + (skel_u64)t * per;
            kt = first >= n ? 0 : ((n - first) < per ? (n - first) : per);
            for (skel_u64 k = 0; k < kt; ++k) {
                VT e;
                e.v = in[first + k];
                e.ok = true;
                mine = comb(mine, e, tup);
            }
        }
        cons_sync();  // the last tile's readers of wsc are done
        VT tot;
        const VT excl = cons_exscan1(mine, wsc[0], tot, tup);
        const VT pre = comb(carry_end, excl, tup);
        skel_T r = pre.v;  // second pass (in-place safe: read, then write)
        for (skel_u64 k = 0; k < kt; ++k) {
            const skel_T e = in[first + k];
            out[first + k] = r;
            r = opf(r, e, tup);
        }
        if (t == 0 && total) total->v = comb(carry_end, tot, tup).v;
    }
    cons_sync();
    if (t == 0) {
        __threadfence();
        const unsigned prev = atomicAdd(&counters[1], 1u);
        if (prev == gridDim.x - 1) {
            counters[1] = 0;
            *epoch_ptr = epoch >= (1u << 30) - 1 ? 1u : epoch + 1;
            __threadfence();
        }
    }
}

// ============================================================================
// Scan for small vectors: two short launches instead of the
// persistent pipeline, whose fixed costs (per-CTA prologue, a 64 KB tile per
// CTA, one status poll round trip per slice) dominate below a few MB.
//   skel_scan_agg_kernel:   aggregate of every tile of RB x SPER elements
//   skel_scan_small_kernel: per tile, prefix = carry (+) aggregates of the
//                           tiles before it (ordered block fold), then an
//                           ordered in-tile exclusive scan
// The second read of the input hits L2 at these sizes (12 B/element of L2/HBM
// traffic instead of 8); in-place is safe (a CTA reads its tile before any of
// its threads writes).
// ============================================================================
constexpr int SPER = SKEL_SCAN_SPER;  // elements per thread
constexpr skel_u64 SM_TILE = (skel_u64)RB * SPER;
constexpr bool SVEC = TMA_OK && (SPER * sizeof(skel_T)) % 16 == 0;

// this thread's SPER contiguous elements from index i0 (valid: i0 + k < n)
template <int PER = SPER>
__device__ __forceinline__ int small_load(const skel_T *in, skel_u64 n, skel_u64 i0, skel_T *x) {
    constexpr bool VEC = TMA_OK && (PER * sizeof(skel_T)) % 16 == 0;
    if (i0 >= n) return 0;
    const skel_u64 left = n - i0;
    if constexpr (VEC) {
        if (left >= (skel_u64)PER && ((reinterpret_cast<unsigned long long>(in + i0) & 15ull) == 0)) {
            constexpr int NQ = skel::cmax<int>(1, (int)(PER * sizeof(skel_T) / 16));
            skel::arr<uint4, NQ> q;
            const uint4 *p = reinterpret_cast<const uint4 *>(in + i0);
#pragma unroll
            for (int j = 0; j < NQ; ++j) q.v[j] = __ldg(p + j);
            const auto e = skel::bit_cast<skel::arr<skel_T, PER>>(q);
#pragma unroll
            for (int k = 0; k < PER; ++k) x[k] = e.v[k];
            return PER;
        }
    }
    const int m = left < (skel_u64)PER ? (int)left : PER;
#pragma unroll
    for (int k = 0; k < PER; ++k)
        if (k < m) x[k] = in[i0 + k];
    return m;
}

// ordered fold of one tile of RB x PER elements into aggs[blockIdx.x]
template <int PER, class Tup>
__device__ __forceinline__ void tile_aggregate(const skel_T *in, skel_u64 n, skel_S *aggs, VT *wpart, Tup &tup,
                                               bool EARLY_TRIGGER) {
    const int t = threadIdx.x;
    skel_T x[PER];
    const int m = small_load<PER>(in, n, blockIdx.x * ((skel_u64)RB * PER) + (skel_u64)t * PER, x);
    // the dependent launch (it waits for our stores) may start: the Reduce's
    // one-CTA fold as soon as the tiles are loaded; the tile Scan, whose CTAs
    // would take SM slots from ours, only once every aggregate is out
    if (EARLY_TRIGGER) skel::pdl_trigger();
    VT a;
    a.ok = false;
#pragma unroll
    for (int k = 0; k < PER; ++k)
        if (k < m) a = comb(a, vt_make(x[k]), tup);
    const VT r = block_fold(a, wpart, tup);
    if (t == 0) aggs[blockIdx.x].v = r.v;  // every tile holds >= 1 element
    if (!EARLY_TRIGGER) skel::pdl_trigger();
}

// (`early`: the dependent kernel is the Reduce's fold, else the tile Scan)
extern "C" __global__ void __launch_bounds__(RB)
    skel_scan_agg_kernel(const skel_T *__restrict__ in, skel_u64 n, skel_S *aggs, int early, const skel_Buf args) {
    auto tup = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    __shared__ VT wpart[NW];
    tile_aggregate<SPER>(in, n, aggs, wpart, tup, early != 0);
}
// the same with tiles of twice the size: the small-vector Reduce above 2^21
// 4-byte elements (more bytes in flight per thread)
extern "C" __global__ void __launch_bounds__(RB)
    skel_red_agg2_kernel(const skel_T *__restrict__ in, skel_u64 n, skel_S *aggs, const skel_Buf args) {
    auto tup = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    __shared__ VT wpart[NW];
    tile_aggregate<2 * SPER>(in, n, aggs, wpart, tup, true);
}

extern "C" __global__ void __launch_bounds__(RB)
    skel_scan_small_kernel(const skel_T *in, skel_T *out, skel_u64 n, const skel_S *aggs, const skel_S identity,
                           const skel_S *seed, const skel_Buf args) {
    auto tup = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    __shared__ VT wpart[NW];
    __shared__ VT wsc[NW];
    __shared__ VT s_pre;
    const int t = threadIdx.x;
    const skel_u64 b = blockIdx.x;
    skel_T x[SPER];  // loaded first: its latency overlaps the prefix fold
    const int m = small_load(in, n, b * SM_TILE + (skel_u64)t * SPER, x);
    skel::pdl_wait();  // the tile aggregates (launched as a programmatic dependent of their kernel)
    // prefix of the tiles before this one, folded in order
    const skel_u64 per = (b + RB - 1) / RB;
    VT a;
    a.ok = false;
    for (skel_u64 k = 0; k < per; ++k) {
        const skel_u64 j = (skel_u64)t * per + k;
        if (j < b) a = comb(a, vt_make(aggs[j].v), tup);
    }
    const VT tiles = block_fold(a, wpart, tup);
    if (t == 0) {
        VT carry;
        carry.v = seed ? seed->v : identity.v;  // as the persistent Scan: out[0] = seed or identity
        carry.ok = true;
        s_pre = comb(carry, tiles, tup);
    }
    VT mine;
    mine.ok = false;
#pragma unroll
    for (int k = 0; k < SPER; ++k)
        if (k < m) mine = comb(mine, vt_make(x[k]), tup);
    VT tot;
    const VT excl = block_exscan(mine, wsc, &tot, tup);  // its barriers also publish s_pre
    skel_T r = comb(s_pre, excl, tup).v;
    skel_T *o = out + b * SM_TILE + (skel_u64)t * SPER;
    if constexpr (SVEC) {
        if (m == SPER && ((reinterpret_cast<unsigned long long>(o) & 15ull) == 0)) {  // 128-bit stores
            skel::arr<skel_T, SPER> y;
#pragma unroll
            for (int k = 0; k < SPER; ++k) {
                y.v[k] = r;
                r = opf(r, x[k], tup);
            }
            constexpr int NQ = skel::cmax<int>(1, (int)(SPER * sizeof(skel_T) / 16));
            const auto q = skel::bit_cast<skel::arr<uint4, NQ>>(y);
#pragma unroll
            for (int j = 0; j < NQ; ++j) reinterpret_cast<uint4 *>(o)[j] = q.v[j];
            return;
        }
    }
#pragma unroll
    for (int k = 0; k < SPER; ++k) {
        if (k < m) {
            const skel_T e = x[k];
            o[k] = r;
            r = opf(r, e, tup);
        }
    }
}

// Reduce for small vectors: skel_scan_agg_kernel's tile aggregates, then this
// one-CTA ordered fold of them (two short launches instead of the TMA ring
// and the last-CTA handshake)
extern "C" __global__ void __launch_bounds__(RB)
    skel_fold_aggs_kernel(const skel_S *aggs, skel_u64 count, skel_S *out, const __grid_constant__ skel_xdev xd,
                          const skel_Buf args) {
    auto tup = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    skel::pdl_wait();  // the tile aggregates (programmatic dependent launch)
    __shared__ VT wpart[NW];
    const int t = threadIdx.x;
    const skel_u64 per = (count + RB - 1) / RB;
    VT a;
    a.ok = false;
    for (skel_u64 k0 = 0; k0 < per; k0 += 8) {  // loads in batches of 8, folded in order
        VT e[8];
#pragma unroll
        for (int u = 0; u < 8; ++u) {
            const skel_u64 j = (skel_u64)t * per + k0 + u;
            e[u].ok = k0 + u < per && j < count;
            if (e[u].ok) e[u].v = aggs[j].v;
        }
#pragma unroll
        for (int u = 0; u < 8; ++u) a = comb(a, e[u], tup);
    }
    const VT r = block_fold(a, wpart, tup);
    if (t == 0) {
        out->v = r.v;
        if (xd.K) skel_xdev_finish(xd, r.v, tup);
    }
}
