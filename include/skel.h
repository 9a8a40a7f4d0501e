/*
 * skel.h -- C-ABI of libskel, a B200-native (sm_100a) rebuild of the
 * data-parallel hot path of SkelCL (Steuwer, Kegel, Gorlatch, "SkelCL - A
 * Portable Skeleton Library for High-Level GPU Programming", IPDPS 2011).
 * Citations "P:Lx-y" are lines of /root/reference/PAPER.md; "R<k>" are the
 * readings listed in DESIGN.md §2.
 *
 * Conventions (all entry points):
 *  - Every call returns a skel_status; SKEL_OK == 0.  No C++ exception ever
 *    crosses this boundary.  skel_last_error() returns a human-readable
 *    message for the last failing call on a context (for SKEL_ERR_COMPILE it
 *    contains the NVRTC log).
 *  - Ownership: handles belong to the caller until *_destroy / skel_finalize
 *    (finalize destroys any vectors still alive).  Host pointers passed in are
 *    BORROWED for the duration of the call only (copy-in / copy-out).  The
 *    library owns all device memory and the pinned host mirrors.
 *  - Asynchrony: skeletons and distribution changes are enqueued on the
 *    context's per-device CUDA streams and return immediately.
 *    skel_vector_download, skel_reduce (which returns a host value, like
 *    Scalar::getValue) and skel_sync block.  Asynchronous device
 *    faults surface as SKEL_ERR_CUDA / SKEL_ERR_NCCL at the next blocking call.
 *  - Threading: one host thread drives a context (the paper's single host
 *    program).
 *  - There is no CPU fallback: without a usable CUDA device every compute or
 *    transfer entry point fails with SKEL_ERR_CUDA.
 */
#ifndef SKEL_H
#define SKEL_H

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef struct skel_ctx_s *skel_ctx_t;
typedef struct skel_vec_s *skel_vec_t;

typedef enum {
    SKEL_OK = 0,
    SKEL_ERR_ARG = 1,     /* NULL handle, bad enum, bad argument list           */
    SKEL_ERR_SIZE = 2,    /* length mismatch (Zip), Reduce of n = 0  */
    SKEL_ERR_TYPE = 3,    /* elem_size != sizeof(parameter), vector/scalar kind  */
    SKEL_ERR_COMPILE = 4, /* NVRTC rejected the user function (log in last_error) */
    SKEL_ERR_CUDA = 5,    /* CUDA runtime/driver error (incl. no device)          */
    SKEL_ERR_NCCL = 6,    /* NCCL error in a distribution change                  */
    SKEL_ERR_OOM = 7,     /* device or pinned host allocation failed              */
    SKEL_ERR_STATE = 8    /* call not valid in the vector's/context's state       */
} skel_status;

/* Distributions, P:L348-351 (copy, block) and Listing 4 P:L522-527;
 * SKEL_SINGLE (whole vector on logical device 0) is reading R6. */
typedef enum { SKEL_SINGLE = 0, SKEL_BLOCK = 1, SKEL_COPY = 2 } skel_dist;

/* Element-wise combine applied when leaving SKEL_COPY (Listing 4 P:L543-546:
 * "reduce (element-wise add) all copies").  Requires a numeric dtype. */
typedef enum {
    SKEL_COMBINE_NONE = 0,
    SKEL_COMBINE_ADD = 1,
    SKEL_COMBINE_MIN = 2,
    SKEL_COMBINE_MAX = 3,
    SKEL_COMBINE_PROD = 4
} skel_combine;

/* Element type tag; only needed for combines (opaque vectors hold any
 * user struct). */
typedef enum {
    SKEL_DT_OPAQUE = 0,
    SKEL_DT_F32 = 1,
    SKEL_DT_F64 = 2,
    SKEL_DT_I32 = 3,
    SKEL_DT_U32 = 4,
    SKEL_DT_I64 = 5,
    SKEL_DT_U64 = 6
} skel_dtype;

/* One extra argument of a user function (Arguments, §III-C).
 * kind SCALAR: `data` points to `size` bytes copied by value into the launch
 * (must equal sizeof of the parameter).  kind VECTOR: `vec` is a vector whose
 * device pointer (local part or local copy) is passed; the parameter must be
 * a pointer.  Arguments are matched to parameters in array order. */
typedef enum { SKEL_ARG_SCALAR = 0, SKEL_ARG_VECTOR = 1 } skel_arg_kind;
typedef struct {
    int kind;
    const void *data;
    size_t size;
    skel_vec_t vec;
} skel_arg;

typedef struct {
    uint64_t h2d_bytes, d2h_bytes, h2d_copies, d2h_copies;
    uint64_t d2d_bytes;       /* device-to-device bytes moved by the library's own exchanges */
    uint64_t nccl_bytes;      /* bytes handed to NCCL collectives by this process            */
    uint64_t kernel_launches; /* skeleton + built-in kernels launched                        */
    uint64_t compile_mem_hits, compile_disk_hits, compile_misses;
    double compile_ms;   /* total NVRTC time                                          */
    double disk_load_ms; /* total time loading cubins from the disk cache */
    uint64_t scan_coop_fallbacks; /* persistent Scans that could not be made co-resident
                                     (cooperative launch refused) and ran as two launches */
    uint64_t vmm_allocs;          /* vector buffers allocated through VMM (cuMemCreate)     */
    uint64_t mc_binds;            /* multicast objects bound to a vector's device buffers   */
    uint64_t multimem_launches;   /* fused tails run through NVSwitch multicast (multimem)  */
    uint64_t xdev_reduces;        /* block-distributed Reduces folded across devices in the
                                     Reduce kernels themselves (last arriver, one pass)      */
} skel_stats;

/* ---- context ------------------------------------------------------------
 * skel_init: one process drives `num_devices` logical devices (SkelCL::init,
 * P:L196).  -1 = one per visible GPU.  If num_devices exceeds the number of
 * visible GPUs, logical device d runs on GPU d % ngpu ("virtual devices",
 * DESIGN.md §6); exchanges between logical devices use the library's own
 * copy/combine kernels.
 * skel_init_rank: one process per GPU (rank of world), logical device =
 * rank, exchanges through NCCL.  `nccl_id` is the 128-byte id produced by
 * skel_get_unique_id on rank 0 and shared by the caller (e.g. via
 * torch.distributed); it may be NULL when world == 1.  */
int skel_init(int num_devices, skel_ctx_t *out);
int skel_get_unique_id(void *nccl_id_128);
int skel_init_rank(int rank, int world, int cuda_device, const void *nccl_id_128,
                   skel_ctx_t *out);
int skel_finalize(skel_ctx_t ctx);
/* D = number of logical devices; L = those driven by this process. */
int skel_num_devices(skel_ctx_t ctx, int *D, int *L);
/* The CUDA stream (cudaStream_t) of the l-th local logical device. */
int skel_get_stream(skel_ctx_t ctx, int local_index, void **stream);
/* Optional threads per block for skeleton kernels (work-group size,
 * P:L415-419); 0 = the skeleton's default. */
int skel_set_block_size(skel_ctx_t ctx, int threads);
/* Kernel cache directory; NULL = $SKEL_CACHE_DIR or
 * ~/.cache/skel_b200; "" disables the disk cache. */
int skel_set_cache_dir(skel_ctx_t ctx, const char *dir);
/* Clear the in-memory kernel cache (the disk cache is kept). */
int skel_clear_kernel_cache(skel_ctx_t ctx);
int skel_sync(skel_ctx_t ctx); /* waits for the main streams and every asynchronous download */
int skel_get_stats(skel_ctx_t ctx, skel_stats *out);
int skel_reset_stats(skel_ctx_t ctx);
const char *skel_last_error(skel_ctx_t ctx);
const char *skel_status_string(int status);

/* ---- vectors (§III-A) -----------------------------------------
 * create: n elements of elem_size bytes; device memory is allocated at once
 * and zero-filled (reading R3).  Initial distribution: SINGLE if
 * D == 1, else BLOCK (reading R6(iii)).
 * upload: copy n elements from src into the host mirror; the host copy
 * becomes the valid one and the host->device transfer is deferred until a
 * skeleton needs the data (lazy copying).
 * download: blocking; copies the vector's value to dst, transferring from
 * the devices only if they hold newer data.  A copy-distributed
 * vector is read from logical device 0 (reading R6).
 * host_ptr / mark_host_modified: zero-copy access to the pinned host mirror
 * (the caller writes it and then marks it modified).
 * fill: device-side fill with one element value; all device copies valid.
 * set_distribution: change the distribution; with a combine the
 * source must be SKEL_COPY and the per-device copies are merged element-wise
 * (copy->block + add = reduce-scatter, Listing 4).
 * mark_device_modified: dataOnDevicesModified() of Listing 4 (P:L538-539,
 * P:L574-578) after a user function wrote the vector through an argument. */
int skel_vector_create(skel_ctx_t ctx, size_t n, size_t elem_size, skel_vec_t *out);
int skel_vector_destroy(skel_vec_t v);
int skel_vector_set_dtype(skel_vec_t v, skel_dtype dt);
int skel_vector_size(skel_vec_t v, size_t *n, size_t *elem_size);
int skel_vector_upload(skel_vec_t v, const void *src, size_t n);
/* upload_part: host data for elements [lo, lo+count) only.  In one-process-
 * per-GPU mode, uploading exactly this process's block part keeps a host
 * mirror of that part only (no full-size host copy per process); otherwise
 * the range is written into the full host copy. */
int skel_vector_upload_part(skel_vec_t v, size_t lo, const void *src, size_t count);
int skel_vector_download(skel_vec_t v, void *dst, size_t n);
/* Download elements [lo, lo + count) into dst (the counterpart of
 * upload_part).  If the host copy is valid and covers the range it is copied
 * from there; otherwise the range is read straight from the device storage
 * that holds it (one D2H per overlapping part; a pinned dst gives the full
 * PCIe/C2C rate) without touching the host mirror.  In rank mode the range
 * must lie in this rank's block part (or the vector must be copy-distributed
 * and not diverged, or single on rank 0), else SKEL_ERR_STATE.  Blocks.
 * SKEL_ERR_SIZE if the range is outside the vector. */
int skel_vector_download_part(skel_vec_t v, size_t lo, void *dst, size_t count);
/* The same without waiting: the device-to-host copies are enqueued on a
 * per-device download stream (after everything already enqueued for v) and
 * the call returns, so they overlap later uploads and kernels.  dst must be
 * pinned host memory (pageable memory makes the copy synchronous) and stay
 * valid and untouched until skel_sync; operations that write v wait for the
 * copy on the device.  Ranges served from a valid host mirror are copied
 * before the call returns. */
int skel_vector_download_part_async(skel_vec_t v, size_t lo, void *dst, size_t count);
int skel_vector_host_ptr(skel_vec_t v, void **host);
int skel_vector_mark_host_modified(skel_vec_t v);
int skel_vector_fill(skel_vec_t v, const void *value);
/* Discard the contents, switch to `dist` without any exchange and fill every
 * device's storage with `value` (e.g. the per-subset zero error image c of
 * LM OSEM, reading R10(i)). */
int skel_vector_fill_dist(skel_vec_t v, skel_dist dist, const void *value);
int skel_vector_set_distribution(skel_vec_t v, skel_dist dist, skel_combine combine);
/* set_distribution_fn: leave SKEL_COPY with a
 * USER-DEFINED element-wise combine instead of the built-in ones.  combine_src
 * is source text of an associative function  T f(T x, T y)  (the last
 * top-level function, as for the skeletons; sizeof(T) = the element size, no
 * further parameters).  The D copies are folded in device order,
 *   result[i] = f(...f(f(copy_0[i], copy_1[i]), copy_2[i])..., copy_{D-1}[i]),
 * so f need not be commutative (P:L283-288 asks only associativity of a
 * customizing operator).  dist = BLOCK: device k folds part k of every copy
 * (peer reads; one process per GPU: part k of every rank is gathered on rank
 * k over NCCL first); SINGLE: device 0 folds the whole copies; COPY: BLOCK then
 * all-gather.  Works on any element type (no dtype needed).
 * Errors: SKEL_ERR_STATE if the vector is not SKEL_COPY; SKEL_ERR_TYPE if f
 * is not T f(T, T) for this element size; SKEL_ERR_COMPILE with the NVRTC log. */
int skel_vector_set_distribution_fn(skel_vec_t v, skel_dist dist, const char *combine_src);
int skel_vector_get_distribution(skel_vec_t v, skel_dist *dist);
int skel_vector_mark_device_modified(skel_vec_t v);
/* Range [lo, hi) of the vector held by logical device d under the current
 * distribution (block: the part; copy/single: whole or empty). */
int skel_vector_part(skel_vec_t v, int d, size_t *lo, size_t *hi);
/* Device pointer + element count held by the l-th local logical device. */
int skel_vector_device_ptr(skel_vec_t v, int local_index, void **ptr, size_t *count);

/* ---- skeletons (§III-B, eqs. (1)-(4)) --------------------------------------
 * `src` is the customizing function as C/CUDA C++ source text;
 * the LAST top-level function definition in it is the entry point, helpers
 * and struct definitions may precede it.  Parameter order: element(s) first,
 * then the Arguments.  The return type is the output element
 * type; `void` is allowed for Map only (side-effect Map).
 * map:    out[i] = f(in[i], args...)               eq. (1)
 * zip:    out[i] = f(a[i], b[i], args...)          eq. (2)
 * reduce: x_0 (+) ... (+) x_{n-1} -> *result_host  eq. (3); (+) must be
 *         associative, need not be commutative; blocking.
 * reduce_to: same, result left on the device in a 1-element vector (non-blocking).
 * scan:   out = [id, x_0, x_0(+)x_1, ...]          eq. (4) P:L297-299 (exclusive);
 *         `identity` points to one element (the id of (+)); in-place allowed.
 * The output vector is resized to the input length and takes the input's
 * distribution; Zip brings `b` to `a`'s distribution first.  Unequal Zip
 * lengths -> SKEL_ERR_SIZE; a size/type mismatch between vectors or scalar
 * arguments and the function's parameters -> SKEL_ERR_TYPE. */
int skel_map(skel_ctx_t ctx, const char *src, skel_vec_t in, skel_vec_t out,
             const skel_arg *args, int nargs);
/* map_index: Map over the index range [0, n) without an
 * input vector: out[i] = f(i, args...), f given as source text whose first
 * parameter is an integer index (4- or 8-byte; a 4-byte index needs
 * n <= 2^31 - 1, else SKEL_ERR_SIZE).  i is the GLOBAL index: under a block
 * distribution of out, device k evaluates its part's indices.  out takes length
 * n and keeps its distribution; out = NULL for a void f (side effects only),
 * which runs over a block partition of [0, n).  Errors as skel_map. */
int skel_map_index(skel_ctx_t ctx, const char *src, size_t n, skel_vec_t out, const skel_arg *args, int nargs);
/* map_lanes: Map (eq. (1)) in which each element is processed by
 * `lanes` consecutive threads of one warp (lanes = 1, 2, 4, 8, 16 or 32).  The
 * user function has the form  R f(T x, int lane, int lanes, args...)  and is
 * called once per (element, lane); it may combine values across the lanes of
 * its element with the prelude's skel_group_sum(v, lanes) (every lane must
 * call it).  out[i] = lane 0's result; out = NULL for a void f.  For elements
 * that are long sequential jobs (an LM OSEM line of response) on
 * parts too small to fill the GPU with one thread per element.  Distribution,
 * ownership and errors as skel_map; lanes outside the set -> SKEL_ERR_ARG. */
int skel_map_lanes(skel_ctx_t ctx, const char *src, skel_vec_t in, skel_vec_t out, int lanes,
                   const skel_arg *args, int nargs);
int skel_zip(skel_ctx_t ctx, const char *src, skel_vec_t a, skel_vec_t b, skel_vec_t out,
             const skel_arg *args, int nargs);
/* Fused form of Listing 4's tail:
 *   b.set_distribution(BLOCK, combine); out = zip(src, a, b); out -> COPY
 * as ONE kernel per device over peer memory: device k combines the D copies of
 * b on its part (peer loads), keeps the combined part of b, applies the Zip
 * function and stores the result into every device's copy of out (peer
 * stores).  b must be SKEL_COPY with a numeric dtype; a is SKEL_COPY or
 * SKEL_BLOCK (out may be a when a is SKEL_COPY).  Afterwards b is SKEL_BLOCK
 * (combined) and out is SKEL_COPY.  One-process-per-GPU contexts reach the
 * peers' buffers through CUDA IPC (opened once per allocation, collectively)
 * and order the kernel between two one-word all-reduce barriers.  With D = 1,
 * more than 16 devices, or inside a capture, the unfused sequence runs. */
int skel_zip_combine(skel_ctx_t ctx, const char *src, skel_vec_t a, skel_vec_t b, skel_combine combine,
                     skel_vec_t out, const skel_arg *args, int nargs);
int skel_reduce(skel_ctx_t ctx, const char *src, skel_vec_t in, void *result_host,
                const skel_arg *args, int nargs);
int skel_reduce_to(skel_ctx_t ctx, const char *src, skel_vec_t in, skel_vec_t result,
                   const skel_arg *args, int nargs);
int skel_scan(skel_ctx_t ctx, const char *src, skel_vec_t in, skel_vec_t out,
              const void *identity, const skel_arg *args, int nargs);

/* ---- CUDA graphs ------------------------------------------------------------
 * capture_begin/end record every skeleton, distribution change and fill issued
 * in between (on all local devices, NCCL collectives included) into a graph;
 * graph_launch replays that device work.  Host-side bookkeeping (lazy
 * transfers, allocations, compilation) happens once, at capture time, so run
 * the sequence eagerly once before capturing it; calls that would block,
 * reallocate or compile inside a capture fail with SKEL_ERR_STATE. */
typedef struct skel_graph_s *skel_graph_t;
int skel_capture_begin(skel_ctx_t ctx);
int skel_capture_end(skel_ctx_t ctx, skel_graph_t *out);
int skel_graph_launch(skel_graph_t graph);
int skel_graph_destroy(skel_graph_t graph);

/* Compile (or fetch from the caches) the kernels of a skeleton without
 * running them; kind = "map" | "zip" | "reduce" | "scan".  Used to move the
 * one-time NVRTC cost out of timed regions. */
int skel_prepare(skel_ctx_t ctx, const char *kind, const char *src);

/* ---- pure host logic (no device needed) -----------------------------------
 * Name of the entry function of a user source (last top-level definition). */
int skel_entry_name(const char *src, char *name, size_t cap);
/* NVRTC-compile a user function into a skeleton (no device needed): returns
 * SKEL_OK or SKEL_ERR_COMPILE; `log` (may be NULL) receives the NVRTC log,
 * *cubin_bytes the size of the sm_100a cubin. */
int skel_compile_check(const char *kind, const char *src, int fmad, char *log, size_t cap,
                       size_t *cubin_bytes);
/* Part k of n elements on D devices: [k*ceil(n/D), min(n,(k+1)*ceil(n/D))) */
int skel_plan_part(size_t n, int D, int k, size_t *lo, size_t *hi);
/* The exchange a distribution change performs (table T1):
 * writes a SKEL_XCHG_* code. */
typedef enum {
    SKEL_XCHG_NONE = 0,           /* same distribution, or host-only data (lazy)   */
    SKEL_XCHG_SCATTER = 1,        /* single -> block                               */
    SKEL_XCHG_BROADCAST = 2,      /* single -> copy                                */
    SKEL_XCHG_GATHER = 3,         /* block -> single                               */
    SKEL_XCHG_ALLGATHER = 4,      /* block -> copy                                 */
    SKEL_XCHG_LOCAL_SLICE = 5,    /* copy -> block (no combine): keep own slice    */
    SKEL_XCHG_REDUCE_SCATTER = 6, /* copy -> block + combine                       */
    SKEL_XCHG_KEEP_ROOT = 7,      /* copy -> single (no combine)                   */
    SKEL_XCHG_REDUCE = 8,         /* copy -> single + combine                      */
    SKEL_XCHG_ALLREDUCE = 9       /* copy -> copy + combine                        */
} skel_xchg;
int skel_plan_exchange(skel_dist from, skel_dist to, skel_combine combine, int *xchg);

#ifdef __cplusplus
}
#endif
#endif /* SKEL_H */
