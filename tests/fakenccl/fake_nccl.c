/*
 * fake_nccl.c -- TEST INFRASTRUCTURE ONLY.  A host-staged stand-in for the
 * NCCL collectives libskel uses, so that its one-process-per-GPU (rank) code
 * path can be exercised with several processes on ONE GPU (real NCCL refuses
 * two ranks on the same device).  LD_PRELOAD it into the ranks.
 *
 * Every collective: synchronize the caller's stream, copy the rank's
 * contribution into its slot of a file-backed shared buffer, barrier, build
 * the result on the host from the slots, copy it to the device, barrier.
 * Semantics follow NCCL's (counts per rank, in-place conventions are
 * trivially honoured because send data are staged before recv is written).
 */
#define _GNU_SOURCE
#include <cuda_runtime.h>
#include <fcntl.h>
#include <nccl.h>
#include <pthread.h>
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>
#include <string.h>
#include <sys/mman.h>
#include <sys/stat.h>
#include <time.h>
#include <unistd.h>

struct ctl {
    volatile int ready;
    pthread_barrier_t bar;
};
struct ncclComm {
    int rank, nranks;
    char base[200];
    struct ctl *ctl;
};

static size_t tsize(ncclDataType_t t) {
    switch (t) {
        case ncclInt8: case ncclUint8: return 1;
        case ncclFloat16: case ncclBfloat16: return 2;
        case ncclInt32: case ncclUint32: case ncclFloat32: return 4;
        default: return 8;
    }
}

ncclResult_t ncclGetUniqueId(ncclUniqueId *id) {
    memset(id, 0, sizeof *id);
    struct timespec ts;
    clock_gettime(CLOCK_REALTIME, &ts);
    snprintf(id->internal, sizeof id->internal, "fake%d_%ld_%ld", (int)getpid(), (long)ts.tv_sec, ts.tv_nsec);
    return ncclSuccess;
}

ncclResult_t ncclCommInitRank(ncclComm_t *comm, int nranks, ncclUniqueId id, int rank) {
    struct ncclComm *c = calloc(1, sizeof *c);
    c->rank = rank;
    c->nranks = nranks;
    snprintf(c->base, sizeof c->base, "/tmp/skelfake_%s", id.internal);
    char path[128];
    snprintf(path, sizeof path, "%s.ctl", c->base);
    int fd = open(path, O_RDWR | O_CREAT, 0600);
    if (fd < 0 || ftruncate(fd, sizeof(struct ctl)) != 0) return ncclSystemError;
    c->ctl = mmap(NULL, sizeof(struct ctl), PROT_READ | PROT_WRITE, MAP_SHARED, fd, 0);
    close(fd);
    if (rank == 0) {
        pthread_barrierattr_t a;
        pthread_barrierattr_init(&a);
        pthread_barrierattr_setpshared(&a, PTHREAD_PROCESS_SHARED);
        pthread_barrier_init(&c->ctl->bar, &a, (unsigned)nranks);
        __sync_synchronize();
        c->ctl->ready = 1;
    } else {
        while (!c->ctl->ready) usleep(1000);
    }
    pthread_barrier_wait(&c->ctl->bar);
    *comm = c;
    return ncclSuccess;
}

ncclResult_t ncclCommDestroy(ncclComm_t comm) {
    pthread_barrier_wait(&comm->ctl->bar);
    munmap(comm->ctl, sizeof(struct ctl));
    free(comm);
    return ncclSuccess;
}
ncclResult_t ncclCommGetAsyncError(ncclComm_t comm, ncclResult_t *e) {
    (void)comm;
    *e = ncclSuccess;
    return ncclSuccess;
}
const char *ncclGetErrorString(ncclResult_t r) { return r == ncclSuccess ? "success (fake)" : "error (fake)"; }

/* shared slots of `bytes` each */
static char *slots(struct ncclComm *c, size_t bytes, int *fd_out) {
    char path[128];
    snprintf(path, sizeof path, "%s.data", c->base);
    int fd = open(path, O_RDWR | O_CREAT, 0600);
    size_t total = bytes * (size_t)c->nranks + 64;
    struct stat st;
    fstat(fd, &st);
    if ((size_t)st.st_size < total && ftruncate(fd, (off_t)total) != 0) return NULL;
    char *p = mmap(NULL, total, PROT_READ | PROT_WRITE, MAP_SHARED, fd, 0);
    *fd_out = fd;
    return p == MAP_FAILED ? NULL : p;
}

static void combine(void *acc, const void *x, size_t count, ncclDataType_t t, ncclRedOp_t op) {
#define LOOP(T)                                                                  \
    {                                                                            \
        T *a = (T *)acc;                                                         \
        const T *b = (const T *)x;                                               \
        for (size_t i = 0; i < count; ++i) {                                     \
            if (op == ncclSum) a[i] = a[i] + b[i];                               \
            else if (op == ncclProd) a[i] = a[i] * b[i];                         \
            else if (op == ncclMin) a[i] = b[i] < a[i] ? b[i] : a[i];            \
            else a[i] = a[i] < b[i] ? b[i] : a[i];                               \
        }                                                                        \
    }
    switch (t) {
        case ncclFloat32: LOOP(float) break;
        case ncclFloat64: LOOP(double) break;
        case ncclInt32: LOOP(int32_t) break;
        case ncclUint32: LOOP(uint32_t) break;
        case ncclInt64: LOOP(int64_t) break;
        case ncclUint64: LOOP(uint64_t) break;
        case ncclInt8: LOOP(int8_t) break;
        default: LOOP(uint8_t) break;
    }
#undef LOOP
}

enum kind { AG, RS, BC, SC, GA, RD, AR };

/* copies are ordered on the caller's stream and completed before returning
 * (a plain cudaMemcpy from pageable memory may return before the DMA ends) */
static cudaError_t xfer(void *dst, const void *src, size_t bytes, enum cudaMemcpyKind k, cudaStream_t s) {
    cudaError_t e = cudaMemcpyAsync(dst, src, bytes, k, s);
    return e != cudaSuccess ? e : cudaStreamSynchronize(s);
}

static ncclResult_t coll(enum kind k, const void *send, void *recv, size_t count, ncclDataType_t t, ncclRedOp_t op,
                         int root, struct ncclComm *c, cudaStream_t s) {
    const size_t es = tsize(t), R = (size_t)c->nranks, r = (size_t)c->rank;
    size_t in_bytes = count * es;                   /* contribution per rank */
    if (k == RS || k == SC) in_bytes = count * es * R; /* RS: send has R parts; SC: root's send */
    if (cudaStreamSynchronize(s) != cudaSuccess) return ncclUnhandledCudaError;
    pthread_barrier_wait(&c->ctl->bar);
    int fd;
    char *sl = slots(c, in_bytes, &fd);
    if (!sl) return ncclSystemError;
    const int contributes = !((k == BC || k == SC) && (int)r != root);
    if (contributes) {
        char *dst = sl + ((k == BC || k == SC) ? 0 : r * in_bytes);
        if (xfer(dst, send, in_bytes, cudaMemcpyDeviceToHost, s) != cudaSuccess) return ncclUnhandledCudaError;
    }
    pthread_barrier_wait(&c->ctl->bar);
    char *tmp = NULL;
    cudaError_t e = cudaSuccess;
    switch (k) {
        case AG:
            e = xfer(recv, sl, R * in_bytes, cudaMemcpyHostToDevice, s);
            break;
        case RS:
            tmp = malloc(count * es);
            memcpy(tmp, sl + r * count * es, count * es);
            for (size_t d = 1; d < R; ++d) combine(tmp, sl + d * in_bytes + r * count * es, count, t, op);
            e = xfer(recv, tmp, count * es, cudaMemcpyHostToDevice, s);
            break;
        case BC:
            e = xfer(recv, sl, in_bytes, cudaMemcpyHostToDevice, s);
            break;
        case SC:
            e = xfer(recv, sl + r * count * es, count * es, cudaMemcpyHostToDevice, s);
            break;
        case GA:
            if ((int)r == root) e = xfer(recv, sl, R * in_bytes, cudaMemcpyHostToDevice, s);
            break;
        case RD:
        case AR:
            if (k == AR || (int)r == root) {
                tmp = malloc(in_bytes);
                memcpy(tmp, sl, in_bytes);
                for (size_t d = 1; d < R; ++d) combine(tmp, sl + d * in_bytes, count, t, op);
                e = xfer(recv, tmp, in_bytes, cudaMemcpyHostToDevice, s);
            }
            break;
    }
    free(tmp);
    pthread_barrier_wait(&c->ctl->bar);
    munmap(sl, in_bytes * R + 64);
    close(fd);
    return e == cudaSuccess ? ncclSuccess : ncclUnhandledCudaError;
}

ncclResult_t ncclAllGather(const void *s, void *r, size_t n, ncclDataType_t t, ncclComm_t c, cudaStream_t st) {
    return coll(AG, s, r, n, t, ncclSum, 0, c, st);
}
ncclResult_t ncclReduceScatter(const void *s, void *r, size_t n, ncclDataType_t t, ncclRedOp_t op, ncclComm_t c,
                               cudaStream_t st) {
    return coll(RS, s, r, n, t, op, 0, c, st);
}
ncclResult_t ncclBroadcast(const void *s, void *r, size_t n, ncclDataType_t t, int root, ncclComm_t c, cudaStream_t st) {
    return coll(BC, s, r, n, t, ncclSum, root, c, st);
}
ncclResult_t ncclScatter(const void *s, void *r, size_t n, ncclDataType_t t, int root, ncclComm_t c, cudaStream_t st) {
    return coll(SC, s, r, n, t, ncclSum, root, c, st);
}
ncclResult_t ncclGather(const void *s, void *r, size_t n, ncclDataType_t t, int root, ncclComm_t c, cudaStream_t st) {
    return coll(GA, s, r, n, t, ncclSum, root, c, st);
}
ncclResult_t ncclReduce(const void *s, void *r, size_t n, ncclDataType_t t, ncclRedOp_t op, int root, ncclComm_t c,
                        cudaStream_t st) {
    return coll(RD, s, r, n, t, op, root, c, st);
}
ncclResult_t ncclAllReduce(const void *s, void *r, size_t n, ncclDataType_t t, ncclRedOp_t op, ncclComm_t c,
                           cudaStream_t st) {
    return coll(AR, s, r, n, t, op, 0, c, st);
}

/* Symmetric-window API (SKEL_NCCL_WINDOWS=1): not available in this stand-in,
 * so libskel takes its CUDA-IPC path -- the tests check that fallback. */
ncclResult_t ncclMemAlloc(void **ptr, size_t size) {
    (void)size;
    if (ptr) *ptr = NULL;
    return ncclInvalidUsage;
}
ncclResult_t ncclMemFree(void *ptr) {
    (void)ptr;
    return ncclSuccess;
}
ncclResult_t ncclCommWindowRegister(ncclComm_t comm, void *buff, size_t size, ncclWindow_t *win, int flags) {
    (void)comm; (void)buff; (void)size; (void)flags;
    if (win) *win = NULL;
    return ncclInvalidUsage;
}
ncclResult_t ncclCommWindowDeregister(ncclComm_t comm, ncclWindow_t win) {
    (void)comm; (void)win;
    return ncclSuccess;
}
