// map.cuh -- Map (eq. (1)) and Zip (eq. (2))
// skeleton kernel, instantiated by NVRTC for the user function SKEL_FN.
//
//   SKEL_NIN == 1:  out[i] = SKEL_FN(a[i], args...)        (void: side effects only)
//   SKEL_NIN == 2:  out[i] = SKEL_FN(a[i], b[i], args...)
//   SKEL_NIN == 0:  out[i] = SKEL_FN(i, args...)           (index Map over [0, n), NEXT-4;
//                   i is the GLOBAL index, the part's offset is passed in)
//
// B200 mapping (kernel K1): the vector is walked in "chunks" of
// E consecutive elements, E chosen so one chunk of every operand is one
// naturally aligned load/store of <= 16 bytes (LDG.E.128 / STG.E.128 for
// 4-byte elements).  Each thread keeps SKEL_UNROLL chunks in flight
// (grid-stride loop; the grid is sized by the host to a multiple of the SM
// count).  Streaming cache hints (.nc / L1::no_allocate loads, .cs stores)
// keep single-use data from displacing the L2 lines that user functions
// gather through vector arguments.  Elements whose size is not a power of
// two, and unaligned views, take the scalar path.

#ifndef SKEL_NIN
#define SKEL_NIN 1
#endif
#ifndef SKEL_BLOCK
#define SKEL_BLOCK 256
#endif
#ifndef SKEL_UNROLL
#define SKEL_UNROLL 4
#endif

using skel_F = decltype(&SKEL_FN);
using skel_FT = skel::fn<skel_F>;
#ifndef SKEL_LANES
#define SKEL_LANES 0
#endif
// positional (element / index [/ lane, lanes]) parameters
constexpr int SKEL_NPOS = SKEL_NIN == 0 ? 1 : (SKEL_LANES ? SKEL_NIN + 2 : SKEL_NIN);
static_assert(skel_FT::arity >= SKEL_NPOS, "user function has too few parameters for this skeleton");
using skel_A = typename skel_FT::template param<0>;
#if SKEL_NIN == 2
using skel_B = typename skel_FT::template param<1>;
#else
using skel_B = skel_A;
#endif
using skel_R = typename skel_FT::ret;
constexpr bool skel_void = skel::is_void<skel_R>::value;
struct skel_none { unsigned char b; };
template <bool V, class R> struct skel_out_t { using type = skel::decay_t<R>; };
template <class R> struct skel_out_t<true, R> { using type = skel_none; };
using skel_O = typename skel_out_t<skel_void, skel_R>::type;

using skel_Args = typename skel::drop<SKEL_NPOS, typename skel_FT::params>::type;
using skel_Lay = skel::args_layout<skel_Args>;
constexpr skel_u64 SKEL_ARGBYTES = skel::cmax<skel_u64>(16, skel::align_up(skel_Lay::bytes, 16));
using skel_Buf = skel::argbuf<SKEL_ARGBYTES>;
using skel_Seq = typename skel::make_iseq<skel_Lay::n>::type;

// ---- chunking ------------------------------------------------------------
constexpr skel_u64 skel_szA = SKEL_NIN == 0 ? 1 : sizeof(skel_A);  // the index is not loaded
constexpr skel_u64 skel_szB = (SKEL_NIN == 2) ? sizeof(skel_B) : 1;
constexpr skel_u64 skel_szO = skel_void ? 1 : sizeof(skel_O);
constexpr skel_u64 skel_maxsz = skel::cmax(skel_szA, skel::cmax(skel_szB, skel_szO));
constexpr bool skel_vec_ok = skel::pow2(skel_szA) && skel::pow2(skel_szB) && skel::pow2(skel_szO) && skel_maxsz <= 16;
#ifndef SKEL_ITEMS
constexpr int SKEL_E = skel_vec_ok ? (int)(16 / skel_maxsz) : 1;
#else
constexpr int SKEL_E = skel_vec_ok ? (SKEL_ITEMS < (int)(16 / skel_maxsz) ? SKEL_ITEMS : (int)(16 / skel_maxsz)) : 1;
#endif

// ---- signature table, read back by the host once per loaded module ------
// [0] layout version  [1] NIN  [2] arity  [3] sizeof ret (0 = void)
// [4] sizeof a  [5] sizeof b  [6] #extra args  [7] arg buffer bytes
// [8] E (elements per chunk)  [9] block  [10] chunks in flight per thread  [11..15] reserved
// [16 + 4i ..] extra arg i: size, align, is_pointer, offset
struct skel_sig_t { skel_u64 v[16 + 4 * 32]; };
constexpr skel_sig_t skel_make_sig() {
    skel_sig_t s{};
    s.v[0] = 1;
    s.v[1] = SKEL_NIN;
    s.v[2] = skel_FT::arity;
    s.v[3] = skel_void ? 0 : sizeof(skel_O);
    s.v[4] = sizeof(skel_A);
    s.v[5] = (SKEL_NIN == 2) ? sizeof(skel_B) : 0;
    s.v[6] = skel_Lay::n;
    s.v[7] = SKEL_ARGBYTES;
    s.v[8] = SKEL_E;
    s.v[9] = SKEL_BLOCK;
    s.v[10] = SKEL_UNROLL;
    for (int i = 0; i < skel_Lay::n && i < 32; ++i) {
        s.v[16 + 4 * i] = skel_Lay::size(i);
        s.v[17 + 4 * i] = skel_Lay::align(i);
        s.v[18 + 4 * i] = skel_Lay::isptr(i);
        s.v[19 + 4 * i] = skel_Lay::off(i);
    }
    return s;
}
extern "C" __device__ skel_sig_t skel_sig = skel_make_sig();

// Minimum resident CTAs per SM the element-wise kernels are compiled for (a
// register cap of 65536 / (SKEL_BLOCK * SKEL_MINB) per thread).  A user
// function may set it by defining SKEL_MINB in its text (the text precedes
// this template), e.g. a latency-bound function that wants more warps.
#ifdef SKEL_MINB
#define SKEL_EW_BOUNDS __launch_bounds__(SKEL_BLOCK, SKEL_MINB)
#else
#define SKEL_EW_BOUNDS __launch_bounds__(SKEL_BLOCK)
#endif

// ---- streaming loads / stores of one chunk ---------------------------------
#ifndef SKEL_LD_HINT
#define SKEL_LD_HINT ".nc.L1::no_allocate"
#endif
template <int N> __device__ __forceinline__ skel::chunk<N> skel_ld(const void *p) {
    skel::chunk<N> c;
    if constexpr (N == 16) {
        asm volatile("ld.global" SKEL_LD_HINT ".v4.u32 {%0,%1,%2,%3}, [%4];"
                     : "=r"(c.v.x), "=r"(c.v.y), "=r"(c.v.z), "=r"(c.v.w)
                     : "l"(p));
    } else if constexpr (N == 8) {
        asm volatile("ld.global" SKEL_LD_HINT ".v2.u32 {%0,%1}, [%2];" : "=r"(c.v.x), "=r"(c.v.y) : "l"(p));
    } else if constexpr (N == 4) {
        asm volatile("ld.global" SKEL_LD_HINT ".u32 %0, [%1];" : "=r"(c.v) : "l"(p));
    } else {
        c = *reinterpret_cast<const skel::chunk<N> *>(p);
    }
    return c;
}
#ifndef SKEL_ST_HINT
#define SKEL_ST_HINT ".cs"
#endif
template <int N> __device__ __forceinline__ void skel_st(void *p, const skel::chunk<N> &c) {
    if constexpr (N == 16) {
        asm volatile("st.global" SKEL_ST_HINT ".v4.u32 [%0], {%1,%2,%3,%4};" ::"l"(p), "r"(c.v.x), "r"(c.v.y),
                     "r"(c.v.z), "r"(c.v.w)
                     : "memory");
    } else if constexpr (N == 8) {
        asm volatile("st.global" SKEL_ST_HINT ".v2.u32 [%0], {%1,%2};" ::"l"(p), "r"(c.v.x), "r"(c.v.y) : "memory");
    } else if constexpr (N == 4) {
        asm volatile("st.global" SKEL_ST_HINT ".u32 [%0], %1;" ::"l"(p), "r"(c.v) : "memory");
    } else {
        *reinterpret_cast<skel::chunk<N> *>(p) = c;
    }
}

template <class Tup>
__device__ __forceinline__ void skel_apply_chunk(const skel_A *xa, const skel_B *xb, skel_O *yo, Tup &t) {
#pragma unroll
    for (int e = 0; e < SKEL_E; ++e) {
        if constexpr (skel_void) {
#if SKEL_NIN == 2
            skel::caller<skel_Seq>::call(&SKEL_FN, t, xa[e], xb[e]);
#else
            skel::caller<skel_Seq>::call(&SKEL_FN, t, xa[e]);
#endif
        } else {
#if SKEL_NIN == 2
            yo[e] = skel::caller<skel_Seq>::call(&SKEL_FN, t, xa[e], xb[e]);
#else
            yo[e] = skel::caller<skel_Seq>::call(&SKEL_FN, t, xa[e]);
#endif
        }
    }
}

constexpr int skel_CA = (int)(SKEL_E * skel_szA);
constexpr int skel_CB = (int)(SKEL_E * skel_szB);
constexpr int skel_CO = (int)(SKEL_E * skel_szO);

// one chunk: unpack E elements, apply the user function, pack and store
template <class Tup>
__device__ __forceinline__ void skel_chunk_op(const skel::chunk<skel_CA> &ca, const skel::chunk<skel_CB> &cb, char *po,
                                              Tup &t) {
    auto xa = skel::bit_cast<skel::arr<skel_A, SKEL_E>>(ca);
    skel::arr<skel_B, SKEL_E> xb;
    if constexpr (SKEL_NIN == 2) xb = skel::bit_cast<skel::arr<skel_B, SKEL_E>>(cb);
    skel::arr<skel_O, SKEL_E> yo;
    skel_apply_chunk(xa.v, xb.v, yo.v, t);
    if constexpr (!skel_void) skel_st<skel_CO>(po, skel::bit_cast<skel::chunk<skel_CO>>(yo));
}
// Map over elements no 16-byte chunk covers (E == 1), sizes multiple of 4 up
// to 64 bytes: staged through shared memory (see skel_ew_kernel)
// (power-of-two sizes keep the direct loads: measured slower staged for the
// 16-byte pixel pairs of mandelbrot_pairs, a compute-bound Map)
// A user function may turn the staging off (`#define SKEL_STAGE_ELEMS 0`): the
// LM OSEM error-image Map, whose event load is negligible next to its walk and
// which would pay the staging's registers in occupancy.
#ifndef SKEL_STAGE_ELEMS
#define SKEL_STAGE_ELEMS 1
#endif
constexpr bool skel_stage = SKEL_STAGE_ELEMS && SKEL_NIN == 1 && SKEL_E == 1 && !SKEL_LANES && sizeof(skel_A) >= 8 &&
                            sizeof(skel_A) % 4 == 0 && sizeof(skel_A) <= 64 && !skel::pow2(sizeof(skel_A));
template <bool V = skel_void, class Tup>
__device__ __forceinline__ void skel_one_val(const skel_A &x, skel_O *out, skel_u64 i, Tup &t) {
    if constexpr (V) {
        skel::caller<skel_Seq>::call(&SKEL_FN, t, x);
    } else {
        out[i] = skel::caller<skel_Seq>::call(&SKEL_FN, t, x);
    }
}
template <class Tup>
__device__ __forceinline__ void skel_one(const skel_A *a, const skel_B *b, skel_O *out, skel_u64 i, Tup &t) {
    if constexpr (skel_void) {
#if SKEL_NIN == 2
        skel::caller<skel_Seq>::call(&SKEL_FN, t, a[i], b[i]);
#else
        skel::caller<skel_Seq>::call(&SKEL_FN, t, a[i]);
#endif
    } else {
#if SKEL_NIN == 2
        out[i] = skel::caller<skel_Seq>::call(&SKEL_FN, t, a[i], b[i]);
#else
        out[i] = skel::caller<skel_Seq>::call(&SKEL_FN, t, a[i]);
#endif
    }
}

#if SKEL_LANES
// ---------------------------------------------------------------------------
// lanes Map (skel_map_lanes): element i is processed by `lanes` consecutive
// threads of one warp (lanes = 1, 2, 4, ..., 32), which call
// SKEL_FN(a[i], lane, lanes, args...) with lane = 0..lanes-1 and may combine
// values across the group (skel_group_sum).  Lane 0's result is stored.  A
// warp takes 32/lanes consecutive elements per trip of a warp-uniform
// grid-stride loop, so the lanes of an element are always present together.
// Used where one element is a long sequential job and a launch over the
// elements alone would not fill the GPU (the LM OSEM error-image Map over one
// GPU's part of a subset).
// ---------------------------------------------------------------------------
static_assert(SKEL_NIN == 1, "lanes Map: one input vector");
static_assert(skel::same<skel::decay_t<typename skel_FT::template param<1>>, int>::value &&
                  skel::same<skel::decay_t<typename skel_FT::template param<2>>, int>::value,
              "a lanes Map's user function takes (element, int lane, int lanes, args...)");
template <bool V = skel_void, class Tup>
__device__ __forceinline__ void skel_lanes_one(const skel_A *a, skel_O *out, skel_u64 i, int sub, int lanes, Tup &t) {
    if constexpr (V) {
        skel::caller<skel_Seq>::call(&SKEL_FN, t, a[i], sub, lanes);
    } else {
        const skel_O r = skel::caller<skel_Seq>::call(&SKEL_FN, t, a[i], sub, lanes);
        if (sub == 0) out[i] = r;
    }
}
extern "C" __global__ void SKEL_EW_BOUNDS
    skel_ew_kernel(const skel_A *__restrict__ a, const skel_B *__restrict__ b, skel_O *__restrict__ out, skel_u64 n,
                   int lanes, const skel_Buf args) {
    (void)b;
    skel::pdl_wait();  // launched as a programmatic dependent of the previous kernel (prelude.cuh)
    skel::pdl_trigger();
    auto t = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    const int lane = (int)(threadIdx.x & 31u);
    const int sub = lane & (lanes - 1);
    const skel_u64 per_warp = (skel_u64)(32 / lanes);
    const skel_u64 gw = ((skel_u64)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const skel_u64 wstride = ((skel_u64)gridDim.x * blockDim.x) >> 5;
#pragma unroll 1
    for (skel_u64 base = gw * per_warp; base < n; base += wstride * per_warp) {  // warp-uniform
        const skel_u64 i = base + (skel_u64)(lane / lanes);
        if (i < n) skel_lanes_one(a, out, i, sub, lanes, t);
    }
}
#elif SKEL_NIN == 0
static_assert(skel::is_arith<skel::decay_t<skel_A>>::value, "an index Map's first parameter must be an integer index");
// index Map: element c*E + e of this part is index base + c*E + e; outputs are
// staged per chunk and stored with one 128-bit store, like Map.  (The bodies are
// templates on "void result" so that the discarded branch is never checked.)
template <bool V = skel_void, class Tup>
__device__ __forceinline__ skel_u64 skel_idx_chunks(skel_O *out, skel_u64 n, skel_u64 base, skel_u64 tid,
                                                    skel_u64 stride, Tup &t) {
    using I = skel::decay_t<skel_A>;
    if constexpr (SKEL_E > 1 && !V) {
        const skel_u64 nch = n / SKEL_E;
#pragma unroll 1
        for (skel_u64 c = tid; c < nch; c += stride) {
            skel::arr<skel_O, SKEL_E> yo;
#pragma unroll
            for (int e = 0; e < SKEL_E; ++e) yo.v[e] = skel::caller<skel_Seq>::call(&SKEL_FN, t, (I)(base + c * SKEL_E + e));
            skel_st<skel_CO>(reinterpret_cast<char *>(out) + c * skel_CO, skel::bit_cast<skel::chunk<skel_CO>>(yo));
        }
        return nch * SKEL_E;
    } else {
        return 0;
    }
}
template <bool V = skel_void, class Tup>
__device__ __forceinline__ void skel_idx_one(skel_O *out, skel_u64 i, skel_u64 base, Tup &t) {
    using I = skel::decay_t<skel_A>;
    if constexpr (V) {
        skel::caller<skel_Seq>::call(&SKEL_FN, t, (I)(base + i));
    } else {
        out[i] = skel::caller<skel_Seq>::call(&SKEL_FN, t, (I)(base + i));
    }
}
extern "C" __global__ void SKEL_EW_BOUNDS
    skel_ew_kernel(skel_O *__restrict__ out, skel_u64 n, skel_u64 base, int vec_ok, const skel_Buf args) {
    skel::pdl_wait();
    skel::pdl_trigger();
    auto t = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    const skel_u64 tid = (skel_u64)blockIdx.x * blockDim.x + threadIdx.x;
    const skel_u64 stride = (skel_u64)gridDim.x * blockDim.x;
    const skel_u64 done = vec_ok ? skel_idx_chunks(out, n, base, tid, stride, t) : 0;
#pragma unroll 1
    for (skel_u64 i = done + tid; i < n; i += stride) skel_idx_one(out, i, base, t);
}
#else
// the element-wise body with U chunks in flight per thread (U = U for
// the main kernel; U = 1 for skel_ew_kernel_u1, which needs fewer registers and
// so fits twice the CTAs per SM: the better grid for small vectors, whose
// launch is a single wave -- the grid policy decides, runtime.cpp ew_decide)
template <int U>
__device__ __forceinline__ void skel_ew_body(const skel_A *__restrict__ a, const skel_B *__restrict__ b,
                                             skel_O *__restrict__ out, skel_u64 n, int vec_ok, const skel_Buf &args) {
    // every element-wise kernel is launched as a programmatic dependent of the
    // previous kernel on its stream: it may be scheduled during that kernel's
    // last wave and waits here for its completion (and memory) before touching
    // anything; it lets the next launch be scheduled at once
    skel::pdl_wait();
    skel::pdl_trigger();
    auto t = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    const skel_u64 tid = (skel_u64)blockIdx.x * blockDim.x + threadIdx.x;
    const skel_u64 stride = (skel_u64)gridDim.x * blockDim.x;

    skel_u64 done = 0;  // elements covered by the chunked path
    if (SKEL_E > 1 && vec_ok) {
        const skel_u64 nch = n / SKEL_E;
        done = nch * SKEL_E;
        const char *pa = reinterpret_cast<const char *>(a);
        const char *pb = reinterpret_cast<const char *>(b);
        char *po = reinterpret_cast<char *>(out);
        skel_u64 c = tid;
        // `unroll 1` on the grid-stride loops: unrolling them makes the compiler
        // compute trip counts with a 64-bit division before the first load
        // -- measured better for Map at every size; a Zip streams more bytes per
        // chunk and gains from the compiler's 2x unroll above 2^24 (1.92 -> 1.87 ms
        // at 2^30) more than the prologue costs it (tools/ew_unroll_variants.sh).
        // SKEL_MAIN_UNROLL: the main loop's pragma (tuning hook).
#ifndef SKEL_MAIN_UNROLL
#if SKEL_NIN == 2
#define SKEL_MAIN_UNROLL
#else
#define SKEL_MAIN_UNROLL _Pragma("unroll 1")
#endif
#endif
        if constexpr (U == 1) {  // one chunk in flight: the low-register kernel
#pragma unroll 1
            for (; c < nch; c += stride) {
                const skel::chunk<skel_CA> ca = skel_ld<skel_CA>(pa + c * skel_CA);
                skel::chunk<skel_CB> cb{};
                if constexpr (SKEL_NIN == 2) cb = skel_ld<skel_CB>(pb + c * skel_CB);
                skel_chunk_op(ca, cb, po + c * skel_CO, t);
            }
        } else {
        SKEL_MAIN_UNROLL
        for (; c + (U - 1) * stride < nch; c += U * stride) {
            skel::chunk<skel_CA> ca[U];
            skel::chunk<skel_CB> cb[U];
#pragma unroll
            for (int u = 0; u < U; ++u) {
                ca[u] = skel_ld<skel_CA>(pa + (c + u * stride) * skel_CA);
                if constexpr (SKEL_NIN == 2) cb[u] = skel_ld<skel_CB>(pb + (c + u * stride) * skel_CB);
            }
#pragma unroll
            for (int u = 0; u < U; ++u) {
                skel_chunk_op(ca[u], cb[u], po + (c + u * stride) * skel_CO, t);
            }
        }
        // the < U chunks left to this thread: one predicated round, so
        // their loads are in flight together (a loop would pay one memory round
        // trip per chunk -- what bounded vectors of 2^21..2^23 elements, where a
        // thread holds 2-4 chunks)
        if (c < nch) {
            skel::chunk<skel_CA> ca[U];
            skel::chunk<skel_CB> cb[U];
#pragma unroll
            for (int u = 0; u < U; ++u) {
                if (c + u * stride < nch) {
                    ca[u] = skel_ld<skel_CA>(pa + (c + u * stride) * skel_CA);
                    if constexpr (SKEL_NIN == 2) cb[u] = skel_ld<skel_CB>(pb + (c + u * stride) * skel_CB);
                }
            }
#pragma unroll
            for (int u = 0; u < U; ++u)
                if (c + u * stride < nch) skel_chunk_op(ca[u], cb[u], po + (c + u * stride) * skel_CO, t);
        }
        }  // U > 1
    }
    // Elements of a size no single load covers (a 24-byte LM OSEM event): staged
    // through shared memory.  The CTA
    // copies its tile of blockDim elements with coalesced 16-byte loads, then
    // each thread reads its element from shared memory -- instead of every
    // thread issuing sizeof(A)/4 strided 4-byte loads (measured: a Map over
    // 10^6 events that only reads them took 25 us).  Needs a 16-byte aligned
    // input (vec_ok) and 4-byte multiples; the tail and other types: scalar.
    if constexpr (skel_stage) {
        if (vec_ok) {
            __shared__ __align__(16) unsigned char stage[SKEL_BLOCK * sizeof(skel_A)];
            const skel_u64 tstride = (skel_u64)gridDim.x * SKEL_BLOCK;
#pragma unroll 1
            for (skel_u64 t0 = (skel_u64)blockIdx.x * SKEL_BLOCK; t0 < n; t0 += tstride) {
                const skel_u64 cnt = n - t0 < (skel_u64)SKEL_BLOCK ? n - t0 : (skel_u64)SKEL_BLOCK;
                const skel_u64 bytes = cnt * sizeof(skel_A);
                const char *src = reinterpret_cast<const char *>(a) + t0 * sizeof(skel_A);
                __syncthreads();  // the previous tile has been read
                if ((bytes & 15) == 0 && ((t0 * sizeof(skel_A)) & 15) == 0) {
                    for (skel_u64 o = (skel_u64)threadIdx.x * 16; o < bytes; o += (skel_u64)SKEL_BLOCK * 16)
                        *reinterpret_cast<skel::chunk<16> *>(stage + o) = skel_ld<16>(src + o);
                } else {
                    for (skel_u64 o = (skel_u64)threadIdx.x * 4; o < bytes; o += (skel_u64)SKEL_BLOCK * 4)
                        *reinterpret_cast<skel::chunk<4> *>(stage + o) = skel_ld<4>(src + o);
                }
                __syncthreads();
                if (threadIdx.x < cnt)
                    skel_one_val(*reinterpret_cast<const skel_A *>(stage + threadIdx.x * sizeof(skel_A)), out,
                                 t0 + threadIdx.x, t);
            }
            return;
        }
    }
    // scalar path: the tail, or everything for non-vectorisable element types
#pragma unroll 1
    for (skel_u64 i = done + tid; i < n; i += stride) skel_one(a, b, out, i, t);
}
extern "C" __global__ void SKEL_EW_BOUNDS
    skel_ew_kernel(const skel_A *__restrict__ a, const skel_B *__restrict__ b, skel_O *__restrict__ out, skel_u64 n,
                   int vec_ok, const skel_Buf args) {
    skel_ew_body<SKEL_UNROLL>(a, b, out, n, vec_ok, args);
}
extern "C" __global__ void SKEL_EW_BOUNDS
    skel_ew_kernel_u1(const skel_A *__restrict__ a, const skel_B *__restrict__ b, skel_O *__restrict__ out, skel_u64 n,
                      int vec_ok, const skel_Buf args) {
    skel_ew_body<1>(a, b, out, n, vec_ok, args);
}
#endif  // SKEL_NIN == 0

#if SKEL_NIN == 2
// ---------------------------------------------------------------------------
// Fused copy->block combine + Zip + block->copy (Listing 4
// P:L542-548 as one kernel).  Device k owns part [lo, hi): for each element it
// combines the D copies of b (peer loads over NVLink when the copies live on
// other GPUs), keeps the combined value in its own part of b, applies the Zip
// function to a and the combined b, and stores the result into the part of
// every device's copy of out (peer stores).  Replaces reduce-scatter + Zip +
// all-gather: each byte crosses the interconnect once and no intermediate
// round trip through HBM is needed.
// ---------------------------------------------------------------------------
#define SKEL_MAXDEV 16
struct skel_ptrs { void *p[SKEL_MAXDEV]; };

template <class T> __device__ __forceinline__ T skel_comb_op(T x, T y, int op) {
    if constexpr (skel::is_arith<T>::value) {
        if (op == 1) return x + y;
        if (op == 2) return y < x ? y : x;
        if (op == 3) return x < y ? y : x;
        return x * y;
    } else {
        return x;  // never launched: the host requires a numeric dtype for a combine
    }
}

template <class Tup>
__device__ __forceinline__ void skel_zipcomb_elem(const skel_A &xa, const skel_ptrs &bs, int nsrc, skel_B *bown,
                                                  const skel_ptrs &os, int ndst, skel_u64 i, int op, Tup &t) {
    skel_B acc = static_cast<const skel_B *>(bs.p[0])[i];
    for (int d = 1; d < nsrc; ++d) acc = skel_comb_op(acc, static_cast<const skel_B *>(bs.p[d])[i], op);
    bown[i] = acc;
    if constexpr (!skel_void) {
        const skel_O r = skel::caller<skel_Seq>::call(&SKEL_FN, t, xa, acc);
        for (int d = 0; d < ndst; ++d) static_cast<skel_O *>(os.p[d])[i] = r;
    }
}

extern "C" __global__ void SKEL_EW_BOUNDS
    skel_zipcomb_kernel(const skel_A *__restrict__ a, const skel_ptrs bsrc, int nsrc, skel_B *bown,
                        const skel_ptrs odst, int ndst, skel_u64 n, int op, int vec_ok, const skel_Buf args) {
    skel::pdl_wait();
    skel::pdl_trigger();
    auto t = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    const skel_u64 tid = (skel_u64)blockIdx.x * blockDim.x + threadIdx.x;
    const skel_u64 stride = (skel_u64)gridDim.x * blockDim.x;
    skel_u64 done = 0;
    if constexpr (SKEL_E > 1 && !skel_void) {
        if (vec_ok) {
            const skel_u64 nch = n / SKEL_E;
            done = nch * SKEL_E;
#pragma unroll 1
            for (skel_u64 c = tid; c < nch; c += stride) {
                const auto xa = skel::bit_cast<skel::arr<skel_A, SKEL_E>>(
                    skel_ld<skel_CA>(reinterpret_cast<const char *>(a) + c * skel_CA));
                auto acc = skel::bit_cast<skel::arr<skel_B, SKEL_E>>(
                    *reinterpret_cast<const skel::chunk<skel_CB> *>(static_cast<const char *>(bsrc.p[0]) + c * skel_CB));
                for (int d = 1; d < nsrc; ++d) {
                    const auto y = skel::bit_cast<skel::arr<skel_B, SKEL_E>>(
                        *reinterpret_cast<const skel::chunk<skel_CB> *>(static_cast<const char *>(bsrc.p[d]) + c * skel_CB));
#pragma unroll
                    for (int e = 0; e < SKEL_E; ++e) acc.v[e] = skel_comb_op(acc.v[e], y.v[e], op);
                }
                skel_st<skel_CB>(reinterpret_cast<char *>(bown) + c * skel_CB, skel::bit_cast<skel::chunk<skel_CB>>(acc));
                skel::arr<skel_O, SKEL_E> yo;
                skel_apply_chunk(xa.v, acc.v, yo.v, t);
                const auto co = skel::bit_cast<skel::chunk<skel_CO>>(yo);
                for (int d = 0; d < ndst; ++d) skel_st<skel_CO>(static_cast<char *>(odst.p[d]) + c * skel_CO, co);
            }
        }
    }
#pragma unroll 1
    for (skel_u64 i = done + tid; i < n; i += stride) skel_zipcomb_elem(a[i], bsrc, nsrc, bown, odst, ndst, i, op, t);
}

// ---------------------------------------------------------------------------
// The same fused tail through NVSwitch multicast (NVLS; SURVEY.md §8f NEXT-1 in
// its specified form).  b's D copies and out's D copies are each bound to a
// multicast object, so ONE address reaches the same element on every device:
//   multimem.ld_reduce.add  -- the switch reads the element from all D copies
//                              and returns their sum (the copy->block combine),
//   multimem.st             -- the switch writes the result into all D copies
//                              of out (the block->copy all-gather).
// Device k's kernel walks its part [lo, hi): per 16-byte chunk one
// ld_reduce.v4.f32 of b, the combined chunk kept in its own part of b, the
// Zip function applied, one st.v4 of the result.  Each device moves S/D bytes
// of b in and S/D bytes of out out over NVLink (the switch does the fan-in and
// fan-out), against (D-1)/D x S each way for peer loads/stores.  float32 `+`
// combine and 4-byte outputs only; other types use skel_zipcomb_kernel.
// ---------------------------------------------------------------------------
// (templates on the element types B, O so that nothing is checked for the
// element types the host never launches this kernel with)
template <class B, class O, class Tup>
__device__ __forceinline__ void skel_mm_chunk(const skel_A *a, const float *mcb, B *bown, float *mco, skel_u64 c,
                                              Tup &t) {
    if constexpr (skel::same<skel::decay_t<B>, float>::value && sizeof(O) == 4 && SKEL_E == 4 && !skel_void) {
        float4 v;
        asm volatile("multimem.ld_reduce.relaxed.sys.global.add.v4.f32 {%0, %1, %2, %3}, [%4];"
                     : "=f"(v.x), "=f"(v.y), "=f"(v.z), "=f"(v.w)
                     : "l"(mcb + 4 * c)
                     : "memory");
        skel::arr<B, 4> acc;
        acc.v[0] = v.x;
        acc.v[1] = v.y;
        acc.v[2] = v.z;
        acc.v[3] = v.w;
        skel_st<16>(reinterpret_cast<char *>(bown) + c * 16, skel::bit_cast<skel::chunk<16>>(acc));
        const auto xa = skel::bit_cast<skel::arr<skel_A, 4>>(skel_ld<skel_CA>(reinterpret_cast<const char *>(a) + c * skel_CA));
        skel::arr<O, 4> yo;
        skel_apply_chunk(xa.v, acc.v, yo.v, t);
        const auto r = skel::bit_cast<float4>(yo);
        asm volatile("multimem.st.relaxed.sys.global.v4.f32 [%0], {%1, %2, %3, %4};" ::"l"(mco + 4 * c), "f"(r.x),
                     "f"(r.y), "f"(r.z), "f"(r.w)
                     : "memory");
    }
}
template <class B, class O, class Tup>
__device__ __forceinline__ void skel_mm_one(const skel_A *a, const float *mcb, B *bown, float *mco, skel_u64 i,
                                            Tup &t) {
    if constexpr (skel::same<skel::decay_t<B>, float>::value && sizeof(O) == 4 && !skel_void) {
        float v;
        asm volatile("multimem.ld_reduce.relaxed.sys.global.add.f32 %0, [%1];" : "=f"(v) : "l"(mcb + i) : "memory");
        bown[i] = v;
        const O r = skel::caller<skel_Seq>::call(&SKEL_FN, t, a[i], v);
        asm volatile("multimem.st.relaxed.sys.global.f32 [%0], %1;" ::"l"(mco + i), "f"(skel::bit_cast<float>(r))
                     : "memory");
    }
}
extern "C" __global__ void SKEL_EW_BOUNDS
    skel_zipcomb_mm_kernel(const skel_A *__restrict__ a, const float *mcb, skel_B *bown, float *mco, skel_u64 n,
                           int vec_ok, const skel_Buf args) {
    skel::pdl_wait();
    skel::pdl_trigger();
    auto t = skel::unpack<skel_Args, skel_Lay, skel_Seq>::run(args);
    const skel_u64 tid = (skel_u64)blockIdx.x * blockDim.x + threadIdx.x;
    const skel_u64 stride = (skel_u64)gridDim.x * blockDim.x;
    skel_u64 nch = 0;  // 16-byte chunks (all pointers aligned)
    if constexpr (SKEL_E == 4) {
        nch = vec_ok ? n / 4 : 0;
#pragma unroll 1
        for (skel_u64 c = tid; c < nch; c += stride) skel_mm_chunk<skel_B, skel_O>(a, mcb, bown, mco, c, t);
    }
#pragma unroll 1
    for (skel_u64 i = nch * 4 + tid; i < n; i += stride) skel_mm_one<skel_B, skel_O>(a, mcb, bown, mco, i, t);
}
#endif
