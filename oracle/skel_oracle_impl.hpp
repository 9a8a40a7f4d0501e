// skel_oracle_impl.hpp -- TEST INFRASTRUCTURE ONLY (see oracle_core.c header).
//
// Sequential definitions of the four SkelCL skeletons (§III-B),
// instantiated for a user function given as source text.  The
// oracle compiles  <prelude> + <user source> + <this header> + <entry points>
// with g++ -O2 -ffp-contract=off -fno-fast-math and runs the loops below one
// element at a time, in index order.  Nothing here is shared with the CUDA
// path.
//
//   map    eq. (1):      out[i] = f(x_i, args...)      (void f: side effects only)
//   zip    eq. (2):  out[i] = f(x_i, y_i, args...)
//   reduce eq. (3):      x_0 (+) x_1 (+) ... (+) x_{n-1}   as a left fold
//   scan   eq. (4):  [id, x_0, x_0(+)x_1, ..., x_0(+)...(+)x_{n-2}]
//
// Arguments (§III-C): extra parameters follow the element(s) in
// push order; a pointer parameter receives a host array (a "vector"
// argument), any other parameter receives a copy of the pushed bytes.
#pragma once
#include <cstddef>
#include <cstdint>
#include <cstring>
#include <tuple>
#include <type_traits>
#include <utility>

namespace skel_oracle {

template <class T>
static T take_arg(void *p) {
    if constexpr (std::is_pointer_v<T>) {
        return reinterpret_cast<T>(p);
    } else {
        T v;
        std::memcpy(&v, p, sizeof(T));
        return v;
    }
}

template <class T>
static size_t arg_size() {
    if constexpr (std::is_pointer_v<T>) return 0;  // vector argument
    else return sizeof(T);
}

template <class R, class... P>
struct sig {
    static void sizes(size_t *out, int *nparams) {
        size_t s[] = {0, arg_size<std::decay_t<P>>()...};
        if constexpr (!std::is_void_v<R>) s[0] = sizeof(R);
        *nparams = (int)sizeof...(P);
        for (int i = 0; i <= (int)sizeof...(P); ++i) out[i] = s[i];
    }
};

// ---- map ---------------------------------------------------------------
template <class R, class X, class... A, size_t... I>
static void map_loop(R (*f)(X, A...), const void *in, void *out, size_t n, void **args,
                     std::index_sequence<I...>) {
    using Xd = std::decay_t<X>;
    std::tuple<std::decay_t<A>...> a{take_arg<std::decay_t<A>>(args[I])...};
    const Xd *x = static_cast<const Xd *>(in);
    for (size_t i = 0; i < n; ++i) {
        if constexpr (std::is_void_v<R>) f(x[i], std::get<I>(a)...);
        else static_cast<R *>(out)[i] = f(x[i], std::get<I>(a)...);
    }
}
template <class R, class X, class... A>
static void map(R (*f)(X, A...), const void *in, void *out, size_t n, void **args) {
    map_loop(f, in, out, n, args, std::index_sequence_for<A...>{});
}

// ---- zip ---------------------------------------------------------------
template <class R, class X, class Y, class... A, size_t... I>
static void zip_loop(R (*f)(X, Y, A...), const void *ina, const void *inb, void *out, size_t n,
                     void **args, std::index_sequence<I...>) {
    using Xd = std::decay_t<X>;
    using Yd = std::decay_t<Y>;
    std::tuple<std::decay_t<A>...> a{take_arg<std::decay_t<A>>(args[I])...};
    const Xd *x = static_cast<const Xd *>(ina);
    const Yd *y = static_cast<const Yd *>(inb);
    for (size_t i = 0; i < n; ++i) {
        if constexpr (std::is_void_v<R>) f(x[i], y[i], std::get<I>(a)...);
        else static_cast<R *>(out)[i] = f(x[i], y[i], std::get<I>(a)...);
    }
}
template <class R, class X, class Y, class... A>
static void zip(R (*f)(X, Y, A...), const void *ina, const void *inb, void *out, size_t n,
                void **args) {
    zip_loop(f, ina, inb, out, n, args, std::index_sequence_for<A...>{});
}

// ---- reduce: left fold (((x0 (+) x1) (+) x2) ... ) -----------------------
template <class R, class X, class Y, class... A, size_t... I>
static void reduce_loop(R (*f)(X, Y, A...), const void *in, void *result, size_t n, void **args,
                        std::index_sequence<I...>) {
    using T = std::decay_t<R>;
    std::tuple<std::decay_t<A>...> a{take_arg<std::decay_t<A>>(args[I])...};
    const T *x = static_cast<const T *>(in);
    T acc = x[0];
    for (size_t i = 1; i < n; ++i) acc = f(acc, x[i], std::get<I>(a)...);
    std::memcpy(result, &acc, sizeof(T));
}
template <class R, class X, class Y, class... A>
static void reduce(R (*f)(X, Y, A...), const void *in, void *result, size_t n, void **args) {
    reduce_loop(f, in, result, n, args, std::index_sequence_for<A...>{});
}

// ---- scan: exclusive, out[0] = id, out[i] = out[i-1] (+) x_{i-1} ----------
template <class R, class X, class Y, class... A, size_t... I>
static void scan_loop(R (*f)(X, Y, A...), const void *in, void *out, size_t n,
                      const void *identity, void **args, std::index_sequence<I...>) {
    using T = std::decay_t<R>;
    std::tuple<std::decay_t<A>...> a{take_arg<std::decay_t<A>>(args[I])...};
    const T *x = static_cast<const T *>(in);
    T *y = static_cast<T *>(out);
    T acc;
    std::memcpy(&acc, identity, sizeof(T));
    for (size_t i = 0; i < n; ++i) {
        y[i] = acc;
        acc = f(acc, x[i], std::get<I>(a)...);
    }
}
template <class R, class X, class Y, class... A>
static void scan(R (*f)(X, Y, A...), const void *in, void *out, size_t n, const void *identity,
                 void **args) {
    scan_loop(f, in, out, n, identity, args, std::index_sequence_for<A...>{});
}

template <class R, class... P>
static void sizes_of(R (*)(P...), size_t *out, int *nparams) {
    sig<R, P...>::sizes(out, nparams);
}

}  // namespace skel_oracle
