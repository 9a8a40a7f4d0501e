// prelude.cuh -- compiled by NVRTC in front of every user function.
//
// SkelCL merges the user's customizing function (a string) with
// the skeleton's own source and compiles the result at run time.
// Here the merge is:  prelude + user source + "#define SKEL_FN <entry>" +
// skeleton template, compiled with -arch=sm_100a -default-device -std=c++17.
// No standard library headers are used: NVRTC compiles this text stand-alone.

// OpenCL address-space qualifiers in user code compile to nothing (a CUDA
// generic pointer reaches global memory).
#define __global
#define __local
#define __private
#define __kernel
#define __constant

typedef unsigned long long skel_u64;
typedef unsigned int skel_u32;
typedef long long skel_i64;

namespace skel {

// ---- minimal type traits ---------------------------------------------------
template <class T> struct rm_ref { using type = T; };
template <class T> struct rm_ref<T &> { using type = T; };
template <class T> struct rm_ref<T &&> { using type = T; };
template <class T> struct rm_cv { using type = T; };
template <class T> struct rm_cv<const T> { using type = T; };
template <class T> struct rm_cv<volatile T> { using type = T; };
template <class T> struct rm_cv<const volatile T> { using type = T; };
template <class T> using decay_t = typename rm_cv<typename rm_ref<T>::type>::type;
template <class T> struct is_ptr { static constexpr bool value = false; };
template <class T> struct is_ptr<T *> { static constexpr bool value = true; };
template <class T> struct is_void { static constexpr bool value = false; };
template <> struct is_void<void> { static constexpr bool value = true; };
template <class T> struct is_arith { static constexpr bool value = false; };
template <> struct is_arith<float> { static constexpr bool value = true; };
template <> struct is_arith<double> { static constexpr bool value = true; };
template <> struct is_arith<int> { static constexpr bool value = true; };
template <> struct is_arith<unsigned> { static constexpr bool value = true; };
template <> struct is_arith<long long> { static constexpr bool value = true; };
template <> struct is_arith<unsigned long long> { static constexpr bool value = true; };
template <> struct is_arith<long> { static constexpr bool value = true; };
template <> struct is_arith<unsigned long> { static constexpr bool value = true; };
template <class A, class B> struct same { static constexpr bool value = false; };
template <class A> struct same<A, A> { static constexpr bool value = true; };

template <int I, class... T> struct nth;
template <class H, class... T> struct nth<0, H, T...> { using type = H; };
template <int I, class H, class... T> struct nth<I, H, T...> { using type = typename nth<I - 1, T...>::type; };

template <int... I> struct iseq {};
template <int N, int... I> struct make_iseq : make_iseq<N - 1, N - 1, I...> {};
template <int... I> struct make_iseq<0, I...> { using type = iseq<I...>; };

template <class... T> struct tlist {};

template <class F> struct fn;
template <class R, class... P> struct fn<R (*)(P...)> {
    using ret = R;
    static constexpr int arity = sizeof...(P);
    template <int I> using param = decay_t<typename nth<I, P...>::type>;
    using params = tlist<decay_t<P>...>;
};

// drop the first K types of a list
template <class L> struct tail;
template <class H, class... T> struct tail<tlist<H, T...>> { using type = tlist<T...>; };
template <int K, class L> struct drop { using type = typename drop<K - 1, typename tail<L>::type>::type; };
template <class L> struct drop<0, L> { using type = L; };

template <class T> constexpr T cmax(T a, T b) { return a > b ? a : b; }
constexpr skel_u64 align_up(skel_u64 x, skel_u64 a) { return (x + a - 1) / a * a; }

// ---- Arguments: packed by value into one kernel parameter ----------------
// Layout = a C struct with one member per extra parameter in order (each at
// the next multiple of its alignment).  The host computes the same offsets
// from the sizes/alignments published in skel_sig[].
template <class L> struct args_layout;
template <> struct args_layout<tlist<>> {
    static constexpr int n = 0;
    static constexpr skel_u64 bytes = 0;
    static constexpr skel_u64 off(int) { return 0; }
    static constexpr skel_u64 size(int) { return 0; }
    static constexpr skel_u64 align(int) { return 1; }
    static constexpr skel_u64 isptr(int) { return 0; }
};
template <class... A> struct args_layout<tlist<A...>> {
    static constexpr int n = sizeof...(A);
    static constexpr skel_u64 size(int i) {
        const skel_u64 s[] = {sizeof(A)...};
        return s[i];
    }
    static constexpr skel_u64 align(int i) {
        const skel_u64 s[] = {alignof(A)...};
        return s[i];
    }
    static constexpr skel_u64 isptr(int i) {
        const skel_u64 s[] = {(skel_u64)is_ptr<A>::value...};
        return s[i];
    }
    static constexpr skel_u64 off(int i) {
        skel_u64 o = 0;
        for (int k = 0; k < i; ++k) o = align_up(o, align(k)) + size(k);
        return align_up(o, align(i));
    }
    static constexpr skel_u64 bytes = off(n - 1) + size(n - 1);
};

template <skel_u64 N> struct argbuf {
    alignas(16) unsigned char b[N];
};

template <class T> __device__ __forceinline__ T load_arg(const unsigned char *p) {
    return *reinterpret_cast<const T *>(p);
}

template <class... T> struct tuple;
template <> struct tuple<> {
    __device__ __forceinline__ tuple() {}
};
template <class H, class... T> struct tuple<H, T...> {
    H head;
    tuple<T...> tail;
    __device__ __forceinline__ tuple() {}
    __device__ __forceinline__ tuple(H h, T... t) : head(h), tail(t...) {}
};
template <int I> struct tget {
    template <class H, class... T> __device__ __forceinline__ static auto &get(tuple<H, T...> &t) {
        return tget<I - 1>::get(t.tail);
    }
};
template <> struct tget<0> {
    template <class H, class... T> __device__ __forceinline__ static H &get(tuple<H, T...> &t) { return t.head; }
};

template <class L, class Lay, class Seq> struct unpack;
template <class... A, class Lay, int... I> struct unpack<tlist<A...>, Lay, iseq<I...>> {
    template <class Buf> __device__ __forceinline__ static tuple<A...> run(const Buf &buf) {
        return tuple<A...>(load_arg<A>(buf.b + Lay::off(I))...);
    }
};

// storage slot for a published element value: size a multiple of 4 bytes
template <class T> struct alignas(alignof(T) > 4 ? alignof(T) : 4) slot { T v; };

// register-friendly bit copies (NVRTC has no memcpy builtin)
template <class D, class S> __device__ __forceinline__ D bit_cast(const S &s) {
    static_assert(sizeof(D) == sizeof(S), "bit_cast size mismatch");
    union U { S s; D d; __device__ U() {} } u;
    u.s = s;
    return u.d;
}
template <class T, int N> struct arr { T v[N]; };

// call f(x..., args...) with the unpacked extra arguments
template <class Seq> struct caller;
template <int... I> struct caller<iseq<I...>> {
    template <class F, class Tup, class... X>
    __device__ __forceinline__ static auto call(F f, Tup &t, X... x) -> decltype(f(x..., tget<I>::get(t)...)) {
        return f(x..., tget<I>::get(t)...);
    }
};

// ---- raw chunk types for vectorised (up to 128-bit) global access ----------
constexpr int chunk_align(int n) { return (n & (n - 1)) ? 1 : (n >= 16 ? 16 : n); }
template <int N> struct chunk { alignas(chunk_align(N)) unsigned char b[N]; };
template <> struct chunk<16> { uint4 v; };
template <> struct chunk<8> { uint2 v; };
template <> struct chunk<4> { unsigned v; };

constexpr bool pow2(skel_u64 x) { return x && !(x & (x - 1)); }

// ---- warp shuffles of arbitrary trivially-copyable T --------------------
template <class T> __device__ __forceinline__ T shfl_down(T v, int d) {
    constexpr int W = (int)((sizeof(T) + 3) / 4);
    union U { T t; unsigned w[W]; U() {} } a, b;
    a.t = v;
#pragma unroll
    for (int i = 0; i < W; ++i) b.w[i] = __shfl_down_sync(0xffffffffu, a.w[i], d);
    return b.t;
}
template <class T> __device__ __forceinline__ T shfl_up(T v, int d) {
    constexpr int W = (int)((sizeof(T) + 3) / 4);
    union U { T t; unsigned w[W]; U() {} } a, b;
    a.t = v;
#pragma unroll
    for (int i = 0; i < W; ++i) b.w[i] = __shfl_up_sync(0xffffffffu, a.w[i], d);
    return b.t;
}
template <class T> __device__ __forceinline__ T shfl_idx(T v, int src) {
    constexpr int W = (int)((sizeof(T) + 3) / 4);
    union U { T t; unsigned w[W]; U() {} } a, b;
    a.t = v;
#pragma unroll
    for (int i = 0; i < W; ++i) b.w[i] = __shfl_sync(0xffffffffu, a.w[i], src);
    return b.t;
}

// ---- PTX helpers: mbarrier + bulk async copies (sm_90+, TMA engine) -------
__device__ __forceinline__ unsigned smem_addr(const void *p) {
    return (unsigned)__cvta_generic_to_shared(p);
}
__device__ __forceinline__ void mbar_init(skel_u64 *bar, unsigned count) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_addr(bar)), "r"(count) : "memory");
}
__device__ __forceinline__ void fence_mbar_init() {
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
}
__device__ __forceinline__ void mbar_expect_tx(skel_u64 *bar, unsigned bytes) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_addr(bar)), "r"(bytes)
                 : "memory");
}
__device__ __forceinline__ bool mbar_try_wait(skel_u64 *bar, unsigned phase) {
    unsigned ok;
    asm volatile(
        "{\n .reg .pred p;\n mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n selp.u32 %0, 1, 0, p;\n}\n"
        : "=r"(ok)
        : "r"(smem_addr(bar)), "r"(phase)
        : "memory");
    return ok != 0;
}
__device__ __forceinline__ void mbar_wait(skel_u64 *bar, unsigned phase) {
    while (!mbar_try_wait(bar, phase)) {
    }
}
// global -> shared bulk copy, completion counted on `bar` (bytes % 16 == 0)
__device__ __forceinline__ void bulk_g2s(void *dst_smem, const void *src, unsigned bytes, skel_u64 *bar) {
    asm volatile(
        "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
            smem_addr(dst_smem)),
        "l"(src), "r"(bytes), "r"(smem_addr(bar))
        : "memory");
}
// shared -> global bulk copy (bytes % 16 == 0)
__device__ __forceinline__ void bulk_s2g(void *dst, const void *src_smem, unsigned bytes) {
    asm volatile("cp.async.bulk.global.shared::cta.bulk_group [%0], [%1], %2;" ::"l"(dst), "r"(smem_addr(src_smem)),
                 "r"(bytes)
                 : "memory");
}
__device__ __forceinline__ void bulk_commit() { asm volatile("cp.async.bulk.commit_group;" ::: "memory"); }
__device__ __forceinline__ void bulk_wait_read0() { asm volatile("cp.async.bulk.wait_group.read 0;" ::: "memory"); }
__device__ __forceinline__ void bulk_wait0() { asm volatile("cp.async.bulk.wait_group 0;" ::: "memory"); }
__device__ __forceinline__ void fence_proxy_async() { asm volatile("fence.proxy.async.shared::cta;" ::: "memory"); }

// ---- release/acquire flags for the decoupled look-back (PTX memory model) -
__device__ __forceinline__ void st_release(unsigned *p, unsigned v) {
    asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ unsigned ld_acquire(const unsigned *p) {
    unsigned v;
    asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ unsigned ld_relaxed_u32(const unsigned *p) {
    unsigned v;
    asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ void st_relaxed_u32(unsigned *p, unsigned v) {
    asm volatile("st.relaxed.gpu.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
// element values published through the flags: word-wise relaxed accesses
__device__ __forceinline__ void fence_acq_rel_gpu() { asm volatile("fence.acq_rel.gpu;" ::: "memory"); }
template <class T> __device__ __forceinline__ void st_value(T *p, const T &v) {
    constexpr int W = (int)((sizeof(T) + 3) / 4);
    union U { T t; unsigned w[W]; U() {} } a;
    a.t = v;
    unsigned *q = reinterpret_cast<unsigned *>(p);
#pragma unroll
    for (int i = 0; i < W; ++i) st_relaxed_u32(q + i, a.w[i]);
}
// programmatic dependent launch (the two-launch small-vector Reduce / Scan):
// the second kernel is launched while the first one runs and waits here until
// the first one has completed and its writes are visible; the first one lets
// it be scheduled once every CTA has loaded its tile.  Both are no-ops for a
// kernel launched without the programmatic attribute.
__device__ __forceinline__ void pdl_wait() { asm volatile("griddepcontrol.wait;" ::: "memory"); }
__device__ __forceinline__ void pdl_trigger() { asm volatile("griddepcontrol.launch_dependents;" ::: "memory"); }
// system scope: values and counters that other GPUs read or write over NVLink
// (the cross-device single-pass Reduce, red.cuh skel_xdev_finish)
__device__ __forceinline__ void fence_acq_rel_sys() { asm volatile("fence.acq_rel.sys;" ::: "memory"); }
__device__ __forceinline__ unsigned atom_add_acq_rel_sys(unsigned *p, unsigned v) {
    unsigned r;
    asm volatile("atom.acq_rel.sys.global.add.u32 %0, [%1], %2;" : "=r"(r) : "l"(p), "r"(v) : "memory");
    return r;
}
__device__ __forceinline__ void st_relaxed_sys_u32(unsigned *p, unsigned v) {
    asm volatile("st.relaxed.sys.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ unsigned ld_relaxed_sys_u32(const unsigned *p) {
    unsigned v;
    asm volatile("ld.relaxed.sys.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
    return v;
}
template <class T> __device__ __forceinline__ void st_value_sys(T *p, const T &v) {
    constexpr int W = (int)((sizeof(T) + 3) / 4);
    union U { T t; unsigned w[W]; U() {} } a;
    a.t = v;
    unsigned *q = reinterpret_cast<unsigned *>(p);
#pragma unroll
    for (int i = 0; i < W; ++i) st_relaxed_sys_u32(q + i, a.w[i]);
}
template <class T> __device__ __forceinline__ T ld_value_sys(const T *p) {
    constexpr int W = (int)((sizeof(T) + 3) / 4);
    union U { T t; unsigned w[W]; U() {} } a;
    const unsigned *q = reinterpret_cast<const unsigned *>(p);
#pragma unroll
    for (int i = 0; i < W; ++i) a.w[i] = ld_relaxed_sys_u32(q + i);
    return a.t;
}
template <class T> __device__ __forceinline__ T ld_value(const T *p) {
    constexpr int W = (int)((sizeof(T) + 3) / 4);
    union U { T t; unsigned w[W]; U() {} } a;
    const unsigned *q = reinterpret_cast<const unsigned *>(p);
#pragma unroll
    for (int i = 0; i < W; ++i) a.w[i] = ld_relaxed_u32(q + i);
    return a.t;
}

}  // namespace skel

// ---- lanes Map (skel_map_lanes): the `lanes` consecutive threads that share
// one element.  A user function of a lanes Map receives (element, lane, lanes,
// args...) and may combine values across the element's lanes with these
// (every lane of the group must call them: they are warp shuffles restricted
// to the group's lanes; lanes is a power of two <= 32).
__device__ __forceinline__ unsigned skel_group_mask(int lanes) {
    const unsigned lane = threadIdx.x & 31u;
    return lanes >= 32 ? 0xffffffffu : (((1u << lanes) - 1u) << (lane & ~(unsigned)(lanes - 1)));
}
// sum over the group (butterfly: every lane gets the same value, since each
// step adds the same two operands in every lane and + is commutative)
template <class T> __device__ __forceinline__ T skel_group_sum(T v, int lanes) {
    const unsigned m = skel_group_mask(lanes);
    for (int o = 1; o < lanes; o <<= 1) v += __shfl_xor_sync(m, v, o, lanes);
    return v;
}
