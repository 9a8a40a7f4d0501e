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
//  * Scan: single-pass decoupled look-back (Merrill & Garland) over
//    dynamically ticketed tiles; tile status words carry an epoch so no
//    memset is needed between launches; outputs are staged in the same
//    swizzled smem stage and written by TMA tensor stores (8 B/element).
//  * Element types whose size is not 4, 8 or 16 bytes, unaligned views and
//    the ragged last tile use direct (LDG/STG) loads with the same ordering.

#ifndef SKEL_RBLOCK
#define SKEL_RBLOCK 512
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
constexpr skel_u64 TILE = (skel_u64)RB * K;
constexpr unsigned TILE_BYTES = (unsigned)(TILE * sizeof(skel_T));
constexpr int STAGES = SKEL_STAGES;
constexpr unsigned DSMEM = TMA_OK ? STAGES * TILE_BYTES + 1024 : 0;
// Scan: SRB consumer rows per tile, SSTAGES smem stages
#ifndef SKEL_SCAN_RB
#define SKEL_SCAN_RB 384
#endif
#ifndef SKEL_SCAN_STAGES
#define SKEL_SCAN_STAGES 4
#endif
constexpr int SRB = SKEL_SCAN_RB;
constexpr int SNW = SRB / 32;
constexpr int SSTAGES = SKEL_SCAN_STAGES;
constexpr skel_u64 STILE = (skel_u64)SRB * K;
constexpr unsigned STILE_BYTES = (unsigned)(STILE * sizeof(skel_T));
constexpr unsigned SDSMEM = TMA_OK ? SSTAGES * STILE_BYTES + 1024 : 0;
constexpr bool PACKED = sizeof(skel_S) == 4;  // status = value:32 | epoch:30 | state:2

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
    s.v[14] = SRB + 64;  // scan kernel block size (consumers + producer + look-back warps)
    s.v[15] = STILE;
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
        constexpr int PER = (int)(16 / sizeof(skel_T));
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
        constexpr int PER = (int)(16 / sizeof(skel_T));
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
extern "C" __global__ void __launch_bounds__(RB, 1)
    skel_reduce_kernel(const __grid_constant__ skel_tmap tin, const skel_T *__restrict__ in, skel_u64 n, int use_tma,
                       skel_S *partials, unsigned *pvalid, unsigned *counter, skel_S *result, const skel_Buf args) {
    auto tup = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    __shared__ skel_u64 bars[STAGES];
    __shared__ VT wpart[NW];
    __shared__ int s_last;
    const int t = threadIdx.x;
    const skel_u64 nft = n / TILE;
    const skel_u64 G = gridDim.x, c = blockIdx.x;
    const skel_u64 t0 = nft * c / G, t1 = nft * (c + 1) / G, my = t1 - t0;
    VT run;
    run.ok = false;

    if (TMA_OK && use_tma) {
        unsigned char *stages = aligned_stages(skel_dsmem);
        if (t == 0) {
            for (int s = 0; s < STAGES; ++s) skel::mbar_init(&bars[s], 1);
            skel::fence_mbar_init();
            tma_prefetch_desc(&tin);
        }
        __syncthreads();
        if (t == 0)
            for (skel_u64 s = 0; s < STAGES && s < my; ++s) issue_tile(stages + s * TILE_BYTES, &tin, t0 + s, &bars[s]);
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
            if (t == 0 && i + STAGES < my) issue_tile(stages + s * TILE_BYTES, &tin, t0 + i + STAGES, &bars[s]);
            VT tv = block_fold(a, wpart, tup);
            if (t == 0) run = comb(run, tv, tup);
        }
    } else {
        for (skel_u64 i = 0; i < my; ++i) {
            const skel_T *p = in + (t0 + i) * TILE + (skel_u64)t * K;
            VT a;
            a.v = p[0];
            a.ok = true;
#pragma unroll 4
            for (int k = 1; k < K; ++k) a.v = opf(a.v, p[k], tup);
            __syncthreads();
            VT tv = block_fold(a, wpart, tup);
            if (t == 0) run = comb(run, tv, tup);
        }
    }
    // ragged last tile: direct loads, owned by the last CTA (keeps index order)
    if (c == G - 1 && nft * TILE < n) {
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
        if (t == 0) run = comb(run, tv, tup);
    }
    // publish this CTA's partial; the last CTA to finish folds them in order
    if (t == 0) {
        skel::st_value(&partials[c], skel_S{run.v});
        skel::st_relaxed_u32(&pvalid[c], run.ok ? 1u : 0u);
        __threadfence();
        const unsigned prev = atomicAdd(counter, 1u);
        s_last = (prev == (unsigned)(G - 1));
    }
    __syncthreads();
    if (s_last) {
        __threadfence();
        const skel_u64 per = (G + RB - 1) / RB;
        VT a;
        a.ok = false;
        for (skel_u64 k = 0; k < per; ++k) {
            const skel_u64 j = (skel_u64)t * per + k;
            if (j < G && skel::ld_relaxed_u32(&pvalid[j])) {
                VT e;
                e.v = skel::ld_value(&partials[j]).v;
                e.ok = true;
                a = comb(a, e, tup);
            }
        }
        VT r = block_fold(a, wpart, tup);
        if (t == 0) {
            result->v = r.v;
            *counter = 0;
        }
    }
}

// fold count >= 1 published values in order (cross-device Reduce)
extern "C" __global__ void skel_fold_kernel(const skel_S *vals, int count, skel_S *out, const skel_Buf args) {
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
// Scan (single pass, decoupled look-back, warp-specialised)
//
// CTA = RB consumer threads (one 128-byte row of the tile each) + 1 producer
// warp + 1 look-back warp, one CTA per SM, STAGES smem stages.
//   producer : takes tile tickets (atomic counter), TMA-loads tiles into free
//              stages, and TMA-stores finished stages back to global memory;
//   look-back: as soon as a tile's ticket is known, folds the predecessors'
//              published aggregates / inclusive prefixes (a 256-tile window
//              per round trip), then publishes the tile's inclusive prefix;
//   consumers: in-thread scan of their row, block scan (named barrier 1),
//              publish the tile aggregate, apply the prefix, write the
//              outputs back into the stage.
// Per-stage mbarriers: full (data + ticket), ticket (ticket only), agg
// (tile aggregate ready), prefix (exclusive prefix ready), written
// (outputs in smem, RB arrivals).  Parity of use u of a stage is u & 1.
// ============================================================================
constexpr int SCAN_THREADS = SRB + 64;
constexpr int LB_PER_LANE = 8;  // look-back window = 32 * 8 tiles per round trip

__device__ __forceinline__ void cons_sync() { asm volatile("bar.sync 1, %0;" ::"n"(SRB) : "memory"); }
__device__ __forceinline__ void mbar_arrive(skel_u64 *bar) {
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(skel::smem_addr(bar)) : "memory");
}

// block exclusive scan among the RB consumer threads (named barrier 1)
template <class Tup> __device__ __forceinline__ VT cons_exscan(VT x, VT *wsc, VT *total, Tup &t) {
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
    cons_sync();
    if (w == 0) {
        VT y;
        y.ok = false;
        if (lane < SNW) y = wsc[lane];
        VT yi = y;
#pragma unroll
        for (int d = 1; d < 32; d <<= 1) {
            VT o = vt_shfl_up(yi, d);
            if (lane >= d) yi = comb(o, yi, t);
        }
        VT ye = vt_shfl_up(yi, 1);
        if (lane == 0) ye.ok = false;
        if (lane < SNW) wsc[lane] = ye;
        if (lane == SNW - 1) *total = yi;
    }
    cons_sync();
    return comb(wsc[w], ex, t);
}

__device__ __forceinline__ void publish(skel_u64 *status, unsigned *flags, skel_S *aggv, skel_S *incv, skel_u64 tile,
                                        unsigned epoch, unsigned state, const skel_T &v) {
    if constexpr (PACKED) {
        skel_S sv{v};
        const unsigned bits = skel::bit_cast<unsigned>(sv);
        const skel_u64 word = ((skel_u64)bits << 32) | (skel_u64)((epoch << 2) | state);
        asm volatile("st.release.gpu.global.u64 [%0], %1;" ::"l"(status + tile), "l"(word) : "memory");
    } else {
        skel::st_value(state == 1 ? &aggv[tile] : &incv[tile], skel_S{v});
        skel::st_release(&flags[tile], (epoch << 2) | state);
    }
}
// relaxed read of a tile's status: 0 = not ready, 1 = aggregate, 2 = inclusive
// prefix.  Packed statuses carry their value in the same 64-bit word; for the
// others the value is read after an acquire fence (see read_values).
__device__ __forceinline__ unsigned peek_state(const skel_u64 *status, const unsigned *flags, skel_u64 tile,
                                               unsigned epoch, skel_T &v) {
    if constexpr (PACKED) {
        skel_u64 word;
        asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(word) : "l"(status + tile) : "memory");
        const unsigned lo = (unsigned)word;
        if ((lo >> 2) != epoch) return 0;
        v = skel::bit_cast<skel_S>((unsigned)(word >> 32)).v;
        return lo & 3u;
    } else {
        const unsigned f = skel::ld_relaxed_u32(&flags[tile]);
        if ((f >> 2) != epoch) return 0;
        return f & 3u;
    }
}

extern "C" __global__ void __launch_bounds__(SCAN_THREADS, 1)
    skel_scan_kernel(const __grid_constant__ skel_tmap tin, const __grid_constant__ skel_tmap tout,
                     const skel_T *in, skel_T *out, skel_u64 n, int use_tma, const skel_S identity, const skel_S *seed,
                     skel_u64 *status, unsigned *flags, skel_S *aggv, skel_S *incv, unsigned *counters,
                     unsigned epoch, skel_S *total, const skel_Buf args) {
    auto tup = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    __shared__ skel_u64 full_bar[SSTAGES], tick_bar[SSTAGES], agg_bar[SSTAGES], pre_bar[SSTAGES], wr_bar[SSTAGES];
    __shared__ skel_u64 tq[SSTAGES];
    __shared__ VT s_agg[SSTAGES], s_pre[SSTAGES];
    __shared__ VT wsc[SNW];
    __shared__ VT s_tot;
    const int t = threadIdx.x, lane = t & 31, w = t >> 5;
    const skel_u64 ntiles = (n + STILE - 1) / STILE;
    const bool tma = TMA_OK && use_tma;
    unsigned char *stages = aligned_stages(skel_dsmem);

    if (t == 0) {
        for (int s = 0; s < SSTAGES; ++s) {
            skel::mbar_init(&full_bar[s], 1);
            skel::mbar_init(&tick_bar[s], 1);
            skel::mbar_init(&agg_bar[s], 1);
            skel::mbar_init(&pre_bar[s], 1);
            skel::mbar_init(&wr_bar[s], SRB);
        }
        skel::fence_mbar_init();
    }
    __syncthreads();

    if (w == SNW) {
        // ------------------------------------------------------------ producer
        if (lane == 0) {
            if (tma) {
                tma_prefetch_desc(&tin);
                tma_prefetch_desc(&tout);
            }
            bool done = false;
            skel_u64 last_i = 0;
            for (skel_u64 i = 0;; ++i) {
                const int s = (int)(i % SSTAGES);
                bool stored = false;
                if (i >= SSTAGES) {  // retire the tile that used this stage
                    const skel_u64 old = tq[s];
                    if (old < ntiles) {
                        skel::mbar_wait(&wr_bar[s], (unsigned)(((i / SSTAGES) - 1) & 1));
                        if (tma && (old + 1) * STILE <= n) {
                            const int row = (int)(old * SRB);
                            tma_store_rows(&tout, row, stages + s * STILE_BYTES);
                            tma_store_rows(&tout, row + SRB / 2, stages + s * STILE_BYTES + STILE_BYTES / 2);
                            skel::bulk_commit();
                            stored = true;
                        }
                    }
                }
                // take the ticket only when the stage is about to be refilled (a held
                // ticket delays every later tile's look-back); its latency overlaps
                // the TMA store's read of the stage
                skel_u64 tk = 0;
                if (!done) tk = atomicAdd(&counters[0], 1u);
                if (stored) skel::bulk_wait_read0();
                if (done) {
                    if (i >= last_i + SSTAGES) break;
                    tq[s] = ntiles;
                    continue;
                }
                tq[s] = tk;
                mbar_arrive(&tick_bar[s]);
                if (tk >= ntiles) {
                    done = true;
                    last_i = i;
                    mbar_arrive(&full_bar[s]);
                } else if (tma && (tk + 1) * STILE <= n) {
                    issue_tile<SRB>(stages + s * STILE_BYTES, &tin, tk, &full_bar[s]);
                } else {
                    mbar_arrive(&full_bar[s]);
                }
            }
            skel::bulk_wait0();
        }
    } else if (w == SNW + 1) {
        // ------------------------------------------------------------ look-back
        for (skel_u64 i = 0;; ++i) {
            const int s = (int)(i % SSTAGES);
            const unsigned ph = (unsigned)((i / SSTAGES) & 1);
            skel::mbar_wait(&tick_bar[s], ph);
            const skel_u64 tk = tq[s];
            if (tk >= ntiles) break;
            VT prefix;
            if (tk == 0) {
                prefix.v = seed ? seed->v : identity.v;
                prefix.ok = true;
            } else {
                VT acc;
                acc.ok = false;
                long long j0 = (long long)tk - 1;
                for (;;) {
                    // lane covers tiles j0 - lane*8 - q, q = 0..7 (q = 0 nearest)
                    unsigned st[LB_PER_LANE];
                    skel_T v[LB_PER_LANE];
#pragma unroll
                    for (int q = 0; q < LB_PER_LANE; ++q) {
                        const long long j = j0 - (long long)lane * LB_PER_LANE - q;
                        st[q] = j >= 0 ? peek_state(status, flags, (skel_u64)j, epoch, v[q]) : 3u;
                    }
                    for (;;) {  // re-poll the ones not ready yet
                        bool all = true;
#pragma unroll
                        for (int q = 0; q < LB_PER_LANE; ++q) {
                            if (st[q] == 0) {
                                const long long j = j0 - (long long)lane * LB_PER_LANE - q;
                                st[q] = peek_state(status, flags, (skel_u64)j, epoch, v[q]);
                                all = all && st[q] != 0;
                            }
                        }
                        if (all) break;
                    }
                    if constexpr (!PACKED) {
                        __threadfence();  // acquire: values were published before their flags
#pragma unroll
                        for (int q = 0; q < LB_PER_LANE; ++q) {
                            const long long j = j0 - (long long)lane * LB_PER_LANE - q;
                            if (st[q] == 1) v[q] = skel::ld_value(&aggv[j]).v;
                            if (st[q] == 2) v[q] = skel::ld_value(&incv[j]).v;
                        }
                    }
                    int qp = LB_PER_LANE;  // nearest inclusive prefix of this lane
#pragma unroll
                    for (int q = LB_PER_LANE - 1; q >= 0; --q)
                        if (st[q] == 2) qp = q;
                    const unsigned pm = __ballot_sync(0xffffffffu, qp < LB_PER_LANE);
                    const int lp = pm ? __ffs(pm) - 1 : 32;
                    VT lf;  // lane fold, older (larger q) on the left
                    lf.ok = false;
                    const int qmax = lane < lp ? LB_PER_LANE - 1 : (lane == lp ? qp : -1);
#pragma unroll
                    for (int q = LB_PER_LANE - 1; q >= 0; --q) {
                        if (q <= qmax && st[q] != 3u) {
                            VT e;
                            e.v = v[q];
                            e.ok = true;
                            lf = comb(lf, e, tup);
                        }
                    }
#pragma unroll
                    for (int d = 1; d < 32; d <<= 1) {  // window fold, higher lanes (older) left
                        VT o = vt_shfl_down(lf, d);
                        if ((lane & (2 * d - 1)) == 0) lf = comb(o, lf, tup);
                    }
                    lf = vt_shfl_idx(lf, 0);
                    acc = comb(lf, acc, tup);
                    if (pm) break;
                    j0 -= 32 * LB_PER_LANE;
                }
                prefix = acc;
            }
            skel::mbar_wait(&agg_bar[s], ph);
            const VT agg = s_agg[s];
            const VT inc = comb(prefix, agg, tup);
            if (lane == 0) {
                publish(status, flags, aggv, incv, tk, epoch, 2u, inc.v);
                if (tk == ntiles - 1 && total) total->v = inc.v;
                s_pre[s] = prefix;
                mbar_arrive(&pre_bar[s]);
            }
            __syncwarp();
        }
    } else {
        // ------------------------------------------------------------ consumers
        // iteration i: phase A of tile i (local scan, publish its aggregate),
        // then phase B of tile i-1 (apply its prefix, hand the stage back), so
        // a tile's aggregate is never held up by the previous tile's look-back.
        bool pv = false, pstaged = false;  // previous tile pending phase B
        int ps = 0;
        unsigned pph = 0;
        skel_u64 pfirst = 0, pkt = 0;
        VT pexcl;
        pexcl.ok = false;
        for (skel_u64 i = 0;; ++i) {
            const int s = (int)(i % SSTAGES);
            const unsigned ph = (unsigned)((i / SSTAGES) & 1);
            skel::mbar_wait(&full_bar[s], ph);
            const skel_u64 tk = tq[s];
            const bool live = tk < ntiles;
            if (live) {
                // ---- phase A(i)
                const skel_u64 base = tk * STILE;
                const bool full = base + STILE <= n;
                const bool staged = tma && full;
                VT mine;
                mine.ok = false;
                skel_u64 first = 0, kt = 0;
                skel_T x[K];
                if (staged) {
                    read_row(stages + s * STILE_BYTES, t, x);
#pragma unroll
                    for (int k = 1; k < K; ++k) x[k] = opf(x[k - 1], x[k], tup);
                    mine.v = x[K - 1];
                    mine.ok = true;
                } else {
                    const skel_u64 cnt = full ? STILE : n - base;
                    const skel_u64 per = full ? (skel_u64)K : (cnt + SRB - 1) / SRB;
                    first = base + (skel_u64)t * per;
                    const skel_u64 end = base + cnt;
                    kt = first >= end ? 0 : ((end - first) < per ? (end - first) : per);
                    for (skel_u64 k = 0; k < kt; ++k) {
                        VT e;
                        e.v = in[first + k];
                        e.ok = true;
                        mine = comb(mine, e, tup);
                    }
                }
                const VT excl = cons_exscan(mine, wsc, &s_tot, tup);
                if (t == 0) {
                    const VT tot = s_tot;
                    if (tk > 0) publish(status, flags, aggv, incv, tk, epoch, 1u, tot.v);
                    s_agg[s] = tot;
                    mbar_arrive(&agg_bar[s]);
                }
                if (staged) {
                    // tile-local exclusive results y_k = excl (+) r_{k-1} (y_0 = excl;
                    // row 0 has no excl: its y_0 slot is unused, y_k = r_{k-1})
#pragma unroll
                    for (int k = K - 1; k >= 1; --k) x[k] = excl.ok ? opf(excl.v, x[k - 1], tup) : x[k - 1];
                    x[0] = excl.v;
                    write_row(stages + s * STILE_BYTES, t, x);
                }
                // ---- phase B(i-1)
                if (pv) {
                    skel::mbar_wait(&pre_bar[ps], pph);
                    const VT prefix = s_pre[ps];
                    if (pstaged) {
                        skel_T y[K];
                        read_row(stages + ps * STILE_BYTES, t, y);
#pragma unroll
                        for (int k = 0; k < K; ++k) y[k] = (t == 0 && k == 0) ? prefix.v : opf(prefix.v, y[k], tup);
                        write_row(stages + ps * STILE_BYTES, t, y);
                        skel::fence_proxy_async();
                    } else {
                        const VT pre = comb(prefix, pexcl, tup);
                        skel_T run = pre.v;  // second pass (in-place safe: read, then write)
                        for (skel_u64 k = 0; k < pkt; ++k) {
                            const skel_T e = in[pfirst + k];
                            out[pfirst + k] = run;
                            run = opf(run, e, tup);
                        }
                    }
                    mbar_arrive(&wr_bar[ps]);
                }
                pv = true;
                pstaged = staged;
                ps = s;
                pph = ph;
                pfirst = first;
                pkt = kt;
                pexcl = excl;
            } else {
                // no more tiles: finish the pending one
                if (pv) {
                    skel::mbar_wait(&pre_bar[ps], pph);
                    const VT prefix = s_pre[ps];
                    if (pstaged) {
                        skel_T y[K];
                        read_row(stages + ps * STILE_BYTES, t, y);
#pragma unroll
                        for (int k = 0; k < K; ++k) y[k] = (t == 0 && k == 0) ? prefix.v : opf(prefix.v, y[k], tup);
                        write_row(stages + ps * STILE_BYTES, t, y);
                        skel::fence_proxy_async();
                    } else {
                        const VT pre = comb(prefix, pexcl, tup);
                        skel_T run = pre.v;
                        for (skel_u64 k = 0; k < pkt; ++k) {
                            const skel_T e = in[pfirst + k];
                            out[pfirst + k] = run;
                            run = opf(run, e, tup);
                        }
                    }
                    mbar_arrive(&wr_bar[ps]);
                }
                break;
            }
        }
    }
    __syncthreads();
    if (t == 0) {
        __threadfence();
        const unsigned prev = atomicAdd(&counters[1], 1u);
        if (prev == gridDim.x - 1) {
            counters[0] = 0;
            counters[1] = 0;
        }
    }
}
