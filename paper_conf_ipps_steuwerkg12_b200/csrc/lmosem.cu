// lmosem.cu — context, C ABI (include/lmosem.h) and launch logic of the B200-native
// LM-OSEM subset iteration (§IV, Listings 2-3). Kernels: lmosem_kernels.cuh.
#include <cuda_runtime.h>
#include <nccl.h>
#include <nvtx3/nvToolsExt.h>

#include <fcntl.h>
#include <sys/stat.h>
#include <unistd.h>

#include <algorithm>
#include <cerrno>
#include <chrono>
#include <cmath>
#include <condition_variable>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <mutex>
#include <new>
#include <string>
#include <thread>
#include <vector>

#include "lmosem.h"
#include "lmosem_kernels.cuh"
#include "lmosem_fused.cuh"
#include "lmosem_loop.cuh"

#define LMOSEM_API extern "C" __attribute__((visibility("default")))

namespace {

thread_local std::string g_init_err;  // message of the last failed lmosem_init on this thread

struct PhaseMarks {
    cudaEvent_t e[5];  // start, after f->brick conversion, after project, after combine, after update
};

}  // namespace

#ifndef LMOSEM_FUSED_CTAS_PER_SM
#define LMOSEM_FUSED_CTAS_PER_SM 4  // fused combine: CTAs (and LSA barriers) per SM
#endif

#ifndef LMOSEM_ZLIST
#define LMOSEM_ZLIST 2  // listed z-slab form (lmosem_ctx::zlist_mode)
#endif

#ifndef LMOSEM_WIDE_N
// fused launches of >= this many events use the 28-warp shape (MODE 6). Measured on one
// B200 (profiles/r02_shape_ab): C2 whole subset 0.964 -> 0.947 ms, 1/2 share 0.488 -> 0.487;
// 1/4 and 1/8 shares slower (0.255 -> 0.259, 0.143 -> 0.149): fewer events per warp
#define LMOSEM_WIDE_N 400000
#endif

// reconstruct_host pipelines the final f download in kPipe brick z-ranges
constexpr int kPipe = 8;
// the first subset's upload: kInChunks parts of growing size (1/16, 3/16, 4/16, 8/16 of the
// events). Pinned H2D (~2.3e9 events/s) outruns the projection (~1e9 events/s), so only the
// first, small part's upload is exposed, and few launches keep their ramp/tail cost low.
constexpr int kInChunks = 4;
constexpr int kInChunkEnd[kInChunks + 1] = {0, 1, 4, 8, 16};  // sixteenths of the events

// Loopback group (include/lmosem.h, "Emulated world"): P contexts of one process on one
// GPU act as P ranks. A collective on rank r is a sequence of phases; each phase boundary
// records an event on r's stream, waits at the host barrier for all ranks, then makes r's
// stream wait for every rank's event, so a rank's kernel may read the other ranks' buffers
// exactly when NCCL's collective would have them ready (lmosem_loop.cuh).
struct lmosem_loopback {
    int world = 0;
    int device = -1;
    std::mutex m;
    std::condition_variable cv;
    int arrived = 0;
    uint64_t gen = 0;
    bool broken = false;                 // a rank timed out at a barrier: every later barrier fails
    std::vector<lmosem_ctx*> ranks;      // registered contexts (nullptr = free slot)
    std::vector<const float*> src[2];    // per rank: the buffer published at a phase boundary
                                         // (double-buffered by boundary parity: slot k is rewritten
                                         // only after every rank has passed the next barrier)
    unsigned* bar = nullptr;             // fused combine: device barrier counters (one per CTA index)
    int bar_cap = 0;
};

struct lmosem_ctx {
    int device = -1;
    int32_t dims[3] = {0, 0, 0};
    double vox[3] = {0, 0, 0};
    int64_t V = 0;
    lmk::GridGeom geom{};
    lmk::BrickIt bricks{};
    int64_t nbf = 0;           // floats per padded brick image (8 * bricks)
    int64_t nb_alloc = 0;      // bricks allocated: nb rounded up to a multiple of world
    int combine = 0;           // LMOSEM_COMBINE_* (0 = auto)
    int auto_combine = 0;      // the auto mode: FUSED when multimem set up and self-tested at init, else ISD (world > 1)
    float* c = nullptr;        // error image, bricks (kept all-zero between subsets)
    float* fb = nullptr;       // brick copy of the current f
    float* norm = nullptr;     // s in bricks (halo = 0)
    float* scratch = nullptr;  // V floats, row layout (norm upload)
    int cap = 0;               // path-piece capacity per warp of the full clip box (the largest launch)
    int slabs_forced = 0;      // slab count (0 = automatic from the L2 budget)
    int slab_axis = 2;         // slabs along z, or along the one axis longer than kMaxBox
    int64_t wide_n = LMOSEM_WIDE_N;  // fused launches of at least this many events run MODE 6 (LMOSEM_WIDE_N)
    float* fp_acc = nullptr;   // per-event forward projections of the z-slab passes
    // listed z-slab form (k_zclass): per-launch event lists of a subset
    int zlist_mode = LMOSEM_ZLIST;  // 0: every slab launch runs over all events; 1: coarse lists;
                                    // 2: + fused launches over fine slabs (LMOSEM_ZLIST)
    int zfine_per = 2;         // fine slabs per coarse slab (LMOSEM_ZFINE)
    int zfused_mode = 5;       // k_project mode of the fine-window launches (LMOSEM_ZFUSED_MODE: 5 or 6)
    int zover = 4;             // fine windows overlap: stride = width / zover (LMOSEM_ZOVER)
    int zwin = 0;              // fine window width in voxels (LMOSEM_ZWIN; 0: from zfine_per)
    int zmerge = 1;            // the windows of a coarse slab in one launch (LMOSEM_ZMERGE)
    int zmed = 6;              // medium windows: stride = coarse width / zmed (LMOSEM_ZMED; 0: none)
    int zamerge = 0;           // pass A of all coarse slabs in shared launches (LMOSEM_ZAMERGE)
    int zmwin = 0;             // medium window width in voxels (LMOSEM_ZMWIN; 0: 1.36 x the widest coarse slab)
    int* zlist = nullptr;      // lists, zlist_cap indices each
    int* zcount = nullptr;     // their lengths (kZMaxLists)
    int64_t zlist_cap = 0;
    int zlist_n = 0;           // lists allocated
    unsigned long long* work = nullptr;  // k_project work counters (one per launch in a step)
    int work_next = 0;
    int64_t fp_cap = 0;
    size_t proj_smem = 0;      // dynamic shared memory of k_project
    cudaStream_t own_stream = nullptr, stream = nullptr, copy_stream = nullptr;
    int rank = 0, world = 1;
    ncclComm_t comm = nullptr;
    lmosem_loopback* loop = nullptr;   // loopback transport (test), instead of comm
    cudaEvent_t loop_ev[2] = {nullptr, nullptr};
    int loop_phase = 0;
    const float* loop_peer[lmk::kLoopMax] = {};  // the ranks' buffers published at the last boundary
    bool nccl_mem = false;                          // c, fb from ncclMemAlloc (NVLS-capable)
    void* reg_c = nullptr, * reg_fb = nullptr;       // ncclCommRegister handles
    // fused combine (LMOSEM_COMBINE_FUSED): symmetric windows + device communicator
    ncclWindow_t win_c = nullptr, win_fb = nullptr;
    ncclDevComm dev_comm{};
    bool dev_comm_ok = false, dev_comm_mm = false;
    int fused_ctas = 0;
    int num_sms = 0;
    // programmatic dependent launch (PDL): a kernel enqueued right after one of ours may
    // start its independent prologue (claims, event tiles, float64 LOR setup) while its
    // predecessor drains; it waits (griddepcontrol.wait) before touching f, c or fp.
    // after_kernel: the last operation this library enqueued on `stream` was one of its own
    // kernels (reset by every API entry and every non-kernel operation, so a PDL launch
    // never follows a copy, memset, event, NCCL call or the caller's own work)
    bool pdl = true;
    bool after_kernel = false;
    struct Occ {
        int mode;
        size_t smem;
        int blocks;
    };
    std::vector<Occ> occ;      // k_project residency per (mode, path-buffer bytes)
    bool failed = false;
    std::string err;
    int debug_stall_ms = 0;    // LMOSEM_DEBUG_STALL_MS (tests of the watchdog): a stall before each combine
    int* abort_flag = nullptr; // host-mapped; raised by abort_comm (polled by k_debug_stall)
    // timing
    bool timing = false;
    std::vector<PhaseMarks> pending, pool;
    std::vector<cudaEvent_t> h2d_pending, h2d_pool;
    lmosem_stats st{};
    // host-streaming resources
    lmosem_event* dev_ev[2] = {nullptr, nullptr};
    int64_t dev_ev_cap = 0;
    float* dev_f = nullptr;
    cudaEvent_t ev_copied[2] = {nullptr, nullptr}, ev_consumed[2] = {nullptr, nullptr};
    cudaEvent_t ev_pipe[kPipe + 1] = {};  // host path: per-chunk ready marks (+ f uploaded)
    // file streaming: pinned staging buffers
    lmosem_event* pin_ev[2] = {nullptr, nullptr};
    int64_t pin_cap = 0;
};

namespace {

lmosem_status fail(lmosem_ctx* ctx, lmosem_status s, const std::string& msg) {
    if (ctx) {
        ctx->err = msg;
        if (s == LMOSEM_ECUDA || s == LMOSEM_ENCCL) ctx->failed = true;
    }
    return s;
}

// A buffer the kernels may dereference: device or managed memory, or pinned host memory
// (mapped through UVA). Pageable host memory (cudaMemoryTypeUnregistered) is rejected
// before anything is enqueued, instead of faulting in a kernel and poisoning the context.
bool device_accessible(const void* p) {
    if (!p) return true;  // NULL / empty handled by the callers' own checks
    cudaPointerAttributes a;
    if (cudaPointerGetAttributes(&a, p) != cudaSuccess) {
        (void)cudaGetLastError();
        return false;
    }
    return a.type == cudaMemoryTypeDevice || a.type == cudaMemoryTypeManaged ||
           (a.type == cudaMemoryTypeHost && a.devicePointer != nullptr);
}

bool device_accessible(const void* a, const void* b, const void* c = nullptr) {
    return device_accessible(a) && device_accessible(b) && device_accessible(c);
}

// The event loaders read 8-byte (float2) or, for 16-byte aligned tiles, 16-byte vectors: an
// event array must be 8-byte aligned (every event then is: 24 B records). A misaligned
// pointer is EINVAL before anything is enqueued instead of a kernel fault.
bool events_misaligned(const void* ev, int64_t n) { return n > 0 && ((uintptr_t)ev & 7u) != 0; }

#define CK(call)                                                                                    \
    do {                                                                                            \
        cudaError_t e_ = (call);                                                                    \
        if (e_ != cudaSuccess)                                                                      \
            return fail(ctx, LMOSEM_ECUDA, std::string(#call) + ": " + cudaGetErrorString(e_));     \
    } while (0)

// Allocations: out of memory is ENOMEM and leaves the context usable (the allocation error
// is not sticky and nothing of the failed call has touched c); other errors are ECUDA.
#define CKA(call)                                                                                   \
    do {                                                                                            \
        cudaError_t e_ = (call);                                                                    \
        if (e_ == cudaErrorMemoryAllocation) {                                                      \
            (void)cudaGetLastError();                                                               \
            return fail(ctx, LMOSEM_ENOMEM, std::string(#call) + ": " + cudaGetErrorString(e_));   \
        }                                                                                           \
        if (e_ != cudaSuccess)                                                                      \
            return fail(ctx, LMOSEM_ECUDA, std::string(#call) + ": " + cudaGetErrorString(e_));     \
    } while (0)

#define NK(call)                                                                                    \
    do {                                                                                            \
        ncclResult_t r_ = (call);                                                                   \
        if (r_ != ncclSuccess)                                                                      \
            return fail(ctx, LMOSEM_ENCCL, std::string(#call) + ": " + ncclGetErrorString(r_));     \
    } while (0)

#define USABLE(ctx)                                                                                 \
    do {                                                                                            \
        if (!(ctx)) return LMOSEM_EINVAL;                                                           \
        if ((ctx)->failed) return LMOSEM_ESTATE;                                                    \
        (ctx)->after_kernel = false;                                                                \
    } while (0)

// Launch one of the library's kernels on ctx->stream, as a programmatic dependent launch
// when it directly follows another of ours (see lmosem_ctx::pdl).
template <typename... KArgs, typename... Args>
cudaError_t launch_k(lmosem_ctx* ctx, void (*kernel)(KArgs...), int grid, int block, size_t smem, Args... args) {
    cudaLaunchAttribute at[1];
    at[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    at[0].val.programmaticStreamSerializationAllowed = 1;
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3((unsigned)grid);
    cfg.blockDim = dim3((unsigned)block);
    cfg.dynamicSmemBytes = smem;
    cfg.stream = ctx->stream;
    cfg.attrs = at;
    cfg.numAttrs = (ctx->pdl && ctx->after_kernel) ? 1 : 0;
    const cudaError_t e = cudaLaunchKernelEx(&cfg, kernel, static_cast<KArgs>(args)...);
    ctx->after_kernel = (e == cudaSuccess);
    if (e == cudaSuccess) ctx->st.launches++;
    return e;
}

// LMOSEM_DEBUG_STALL_MS: a bounded spin of `ns` nanoseconds standing in for a peer that is
// late to the combine (tests of the watchdog in wait_done; never set in production). Like
// NCCL's own kernels it also polls an abort flag (host-mapped), which abort_comm raises.
__global__ void k_debug_stall(unsigned long long ns, const volatile int* abort_flag) {
    unsigned long long t0, t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t0));
    do {
        __nanosleep(100000);
        asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    } while (t - t0 < ns && *abort_flag == 0);
}

// any operation on ctx->stream that is not one of the library's kernels
inline void not_kernel(lmosem_ctx* ctx) { ctx->after_kernel = false; }

void block_range(int64_t n, int r, int P, int64_t* b, int64_t* e) {
    // floor(r*n/P) without overflow for n < 2^62 / P
    *b = (int64_t)((__int128)n * r / P);
    *e = (int64_t)((__int128)n * (r + 1) / P);
}

// part q of Q (1: the whole range; kInChunks: the first subset's growing parts) of n events
void in_chunk_range(int64_t n, int q, int Q, int64_t* b, int64_t* e) {
    if (Q == 1) {
        *b = 0;
        *e = n;
        return;
    }
    *b = n * kInChunkEnd[q] / 16;
    *e = n * kInChunkEnd[q + 1] / 16;
}

// ISD combine blocks: the nb bricks are allocated as `alloc` =
// nb rounded up to a multiple of world, split into world equal chunks; rank r owns (reduces,
// updates, all-gathers) chunk r, of which [begin, end) are real bricks (end <= nb)
void isd_block(int64_t nb, int rank, int world, int64_t* begin, int64_t* end, int64_t* alloc) {
    const int64_t a = (nb + world - 1) / world * world;
    const int64_t chunk = a / world;
    *alloc = a;
    *begin = std::min(nb, chunk * rank);
    *end = std::min(nb, chunk * (rank + 1));
}

int grid_for(lmosem_ctx* ctx, int64_t items) {
    const int64_t cap = (int64_t)ctx->num_sms * 16;
    return (int)std::max<int64_t>(1, std::min<int64_t>((items + 255) / 256, cap));
}

int combine_mode(const lmosem_ctx* ctx) {
    if (ctx->combine) return ctx->combine;
    if (ctx->auto_combine) return ctx->auto_combine;
    return ctx->world > 1 ? LMOSEM_COMBINE_ISD : LMOSEM_COMBINE_ALLREDUCE;
}

// ------------------------------------------------------------- the combine's transports
// The collectives of the combine (Listing 3 l.6 copy(add), l.15-16)
// with NCCL's semantics, through the context's transport: NCCL (one process per GPU) or
// the loopback group (P contexts on one GPU; test transport). subset_iteration calls only
// these, so both transports run the same combine code.
bool has_comm(const lmosem_ctx* ctx) { return ctx->comm != nullptr || ctx->loop != nullptr; }

// seconds a host barrier of the loopback group (and lmosem_synchronize on an NCCL context)
// waits before declaring the collective failed (LMOSEM_TIMEOUT_S, default 300)
double coll_timeout_s() {
    const char* e = std::getenv("LMOSEM_TIMEOUT_S");
    const double t = e ? std::atof(e) : 300.0;
    return t > 0 ? t : 300.0;
}

bool loop_barrier(lmosem_loopback* g) {
    std::unique_lock<std::mutex> lk(g->m);
    if (g->broken) return false;
    const uint64_t my = g->gen;
    if (++g->arrived == g->world) {
        g->arrived = 0;
        ++g->gen;
        g->cv.notify_all();
        return true;
    }
    const bool ok = g->cv.wait_for(lk, std::chrono::duration<double>(coll_timeout_s()),
                                   [&] { return g->gen != my || g->broken; });
    if (!ok || g->broken) {
        g->broken = true;
        g->cv.notify_all();
        return false;
    }
    return true;
}

// Phase boundary of a loopback collective on this rank (see lmosem_loopback): publish
// `mine` (read by the other ranks until the next boundary), then order this rank's stream
// after every rank's work so far. Events alternate per boundary, so an event is re-recorded
// only after every rank has passed the barrier that follows its waits on it.
lmosem_status loop_boundary(lmosem_ctx* ctx, const float* mine = nullptr) {
    lmosem_loopback* g = ctx->loop;
    not_kernel(ctx);
    const int ph = ctx->loop_phase;
    CK(cudaEventRecord(ctx->loop_ev[ph], ctx->stream));
    {
        std::lock_guard<std::mutex> lk(g->m);
        g->src[ph][ctx->rank] = mine;
    }
    if (!loop_barrier(g))
        return fail(ctx, LMOSEM_ENCCL, "loopback: a rank did not reach the collective within LMOSEM_TIMEOUT_S");
    {
        std::lock_guard<std::mutex> lk(g->m);
        for (int q = 0; q < ctx->world; ++q) ctx->loop_peer[q] = g->src[ph][q];
    }
    for (int q = 0; q < ctx->world; ++q)
        if (q != ctx->rank) CK(cudaStreamWaitEvent(ctx->stream, g->ranks[q]->loop_ev[ph], 0));
    ctx->loop_phase ^= 1;
    return LMOSEM_OK;
}

lmk::LoopSrc loop_src(const lmosem_ctx* ctx, int64_t add) {
    lmk::LoopSrc src{};
    for (int q = 0; q < ctx->world; ++q) src.p[q] = ctx->loop_peer[q] + add;
    return src;
}

int loop_grid(const lmosem_ctx* ctx, int64_t n) {
    return (int)std::max<int64_t>(1, std::min<int64_t>((n + 255) / 256, (int64_t)ctx->num_sms * 8));
}

// recv[i] = sum over ranks of send[rank * count + i], i < count (send == recv - rank * count: in place)
lmosem_status coll_reduce_scatter(lmosem_ctx* ctx, const float* send, float* recv, size_t count) {
    if (ctx->comm) {
        not_kernel(ctx);
        NK(ncclReduceScatter(send, recv, count, ncclFloat32, ncclSum, ctx->comm, ctx->stream));
        return LMOSEM_OK;
    }
    lmosem_status s;
    if ((s = loop_boundary(ctx, send))) return s;
    const lmk::LoopSrc src = loop_src(ctx, (int64_t)count * ctx->rank);
    lmk::k_loop_sum<<<loop_grid(ctx, (int64_t)count), 256, 0, ctx->stream>>>(src, recv, (int64_t)count, ctx->world);
    CK(cudaGetLastError());
    ctx->st.launches++;
    return loop_boundary(ctx);
}

// recv[rank' * count + i] = send of rank' [i] for every rank' (send == recv + rank * count: in place)
lmosem_status coll_all_gather(lmosem_ctx* ctx, const float* send, float* recv, size_t count) {
    if (ctx->comm) {
        not_kernel(ctx);
        NK(ncclAllGather(send, recv, count, ncclFloat32, ctx->comm, ctx->stream));
        return LMOSEM_OK;
    }
    lmosem_status s;
    if ((s = loop_boundary(ctx, send))) return s;
    lmk::LoopSrc src = loop_src(ctx, 0);
    for (int q = 0; q <= ctx->world; ++q) src.off[q] = (int64_t)count * q;
    dim3 grid((unsigned)loop_grid(ctx, (int64_t)count), (unsigned)ctx->world);
    lmk::k_loop_gather<<<grid, 256, 0, ctx->stream>>>(src, recv, send == recv + (int64_t)count * ctx->rank ? ctx->rank : -1);
    CK(cudaGetLastError());
    ctx->st.launches++;
    return loop_boundary(ctx);
}

// buf <- sum over ranks of buf (in place), count floats
lmosem_status coll_all_reduce(lmosem_ctx* ctx, float* buf, size_t count) {
    if (ctx->comm) {
        not_kernel(ctx);
        NK(ncclAllReduce(buf, buf, count, ncclFloat32, ncclSum, ctx->comm, ctx->stream));
        return LMOSEM_OK;
    }
    // reduce-scatter of block r of the count floats into this rank's buf, then all-gather
    lmk::LoopSrc src{};
    for (int q = 0; q < ctx->world; ++q) block_range((int64_t)count, q, ctx->world, &src.off[q], &src.off[q + 1]);
    const int64_t b = src.off[ctx->rank], n = src.off[ctx->rank + 1] - b;
    lmosem_status s;
    if ((s = loop_boundary(ctx, buf))) return s;
    const lmk::LoopSrc part = loop_src(ctx, b);
    lmk::k_loop_sum<<<loop_grid(ctx, n), 256, 0, ctx->stream>>>(part, buf + b, n, ctx->world);
    CK(cudaGetLastError());
    ctx->st.launches++;
    if ((s = loop_boundary(ctx, buf))) return s;
    for (int q = 0; q < ctx->world; ++q) src.p[q] = ctx->loop_peer[q] + src.off[q];
    dim3 grid((unsigned)loop_grid(ctx, (int64_t)count / ctx->world + 1), (unsigned)ctx->world);
    lmk::k_loop_gather<<<grid, 256, 0, ctx->stream>>>(src, buf, ctx->rank);
    CK(cudaGetLastError());
    ctx->st.launches++;
    return loop_boundary(ctx);
}

// The fused ISD combine (NEXT-1; lmosem_fused.cuh): reduce-scatter of c, the block update
// and the all-gather of f as ONE kernel. NCCL: k_combine_fused over the symmetric windows,
// a programmatic dependent launch after the projection. Loopback: one cooperative launch
// of the same body for all ranks (rank 0 launches it between two phase boundaries).
lmosem_status coll_fused(lmosem_ctx* ctx, int64_t chunk) {
    if (ctx->comm) {
        if (ctx->dev_comm_mm)
            CK(launch_k(ctx, lmk::k_combine_fused<true>, ctx->fused_ctas, 256, 0, ctx->dev_comm, ctx->win_c,
                        ctx->win_fb, (const float*)ctx->norm, ctx->c, (const float*)ctx->fb, chunk, ctx->bricks.nb,
                        ctx->bricks));
        else
            CK(launch_k(ctx, lmk::k_combine_fused<false>, ctx->fused_ctas, 256, 0, ctx->dev_comm, ctx->win_c,
                        ctx->win_fb, (const float*)ctx->norm, ctx->c, (const float*)ctx->fb, chunk, ctx->bricks.nb,
                        ctx->bricks));
        return LMOSEM_OK;
    }
    lmosem_status s;
    if ((s = loop_boundary(ctx))) return s;
    if (ctx->rank == 0) {
        lmosem_loopback* g = ctx->loop;
        const int P = ctx->world;
        int per_sm = 0;
        CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, lmk::k_combine_loop, 256, 0));
        const int ctas = std::max(1, std::min(LMOSEM_FUSED_CTAS_PER_SM * ctx->num_sms, per_sm * ctx->num_sms / P));
        if (ctas > g->bar_cap) {
            if (g->bar) CK(cudaFree(g->bar));
            g->bar = nullptr;
            g->bar_cap = 0;
            CKA(cudaMalloc(&g->bar, sizeof(unsigned) * ctas));
            g->bar_cap = ctas;
        }
        CK(cudaMemsetAsync(g->bar, 0, sizeof(unsigned) * ctas, ctx->stream));
        lmk::LoopImages im{};
        for (int q = 0; q < P; ++q) {
            im.c[q] = g->ranks[q]->c;
            im.fb[q] = g->ranks[q]->fb;
            im.s[q] = g->ranks[q]->norm;
        }
        unsigned* bar = g->bar;
        int64_t nb = ctx->bricks.nb;
        lmk::BrickIt it = ctx->bricks;
        void* args[] = {&im, &bar, (void*)&P, (void*)&ctas, &chunk, &nb, &it};
        CK(cudaLaunchCooperativeKernel((const void*)lmk::k_combine_loop, dim3((unsigned)(P * ctas)), dim3(256), args, 0,
                                       ctx->stream));
        ctx->st.launches++;
    }
    return loop_boundary(ctx);
}

lmosem_status launch_to_brick(lmosem_ctx* ctx, const float* row, float* br) {
    CK(launch_k(ctx, lmk::k_row_to_brick, grid_for(ctx, ctx->bricks.nb), 256, 0, row, br, ctx->geom, ctx->bricks));
    return LMOSEM_OK;
}

lmosem_status launch_to_row(lmosem_ctx* ctx, float* br, float* row, int zero) {
    CK(launch_k(ctx, lmk::k_brick_to_row, grid_for(ctx, ctx->bricks.nb), 256, 0, br, row, ctx->geom, ctx->bricks,
                zero));
    return LMOSEM_OK;
}

// Largest clip-box extent (voxels) whose per-warp path buffer (3 pieces per dominant-axis
// slab, 8 B each) and clip area (768 B), 8 warps per CTA, fit the 227 KB of opt-in shared
// memory of sm_100a.
constexpr int kMaxBox = 1170;

// Largest slab extent along `axis` when it is cut into K even-aligned slabs (slab_geom).
int max_slab_extent(int n_axis, int K) {
    const int half = n_axis / 2;
    int m = 0;
    for (int k = 0; k < K; ++k) {
        const int lo = 2 * (int)((int64_t)half * k / K);
        const int hi = (k == K - 1) ? n_axis : 2 * (int)((int64_t)half * (k + 1) / K);
        m = std::max(m, hi - lo);
    }
    return m;
}

// Number of slabs for the projection, along ctx->slab_axis (z, or the one axis longer than
// kMaxBox): the brick image slab of a pass should stay L2-resident (L2 126 MB; a 72 MB
// budget per image slab leaves room for the event stream and the per-event fp array;
// measured at C4, 208 MB: 2/3/4/5 slabs 27.1/24.5/25.2/26.3 ms), and no slab may be longer
// than kMaxBox along its axis (the path buffer). 1 = the single fused pass.
int n_slabs(const lmosem_ctx* ctx) {
    const int n_axis = ctx->dims[ctx->slab_axis];
    const int max_slabs = std::max(1, n_axis / 2);
    int k_min = 1;  // the path-buffer bound (> 1 only for an axis longer than kMaxBox)
    while (k_min < max_slabs && max_slab_extent(n_axis, k_min) > kMaxBox) ++k_min;
    if (ctx->slabs_forced > 0) return std::max(k_min, std::min(ctx->slabs_forced, max_slabs));
    const double bytes = 4.0 * (double)ctx->nbf;
    const double budget = 72.0 * 1024 * 1024;
    return std::max(k_min, std::min(max_slabs, std::max(1, (int)std::ceil(bytes / budget))));
}

#ifndef LMOSEM_STATIC_BATCH
#define LMOSEM_STATIC_BATCH 1  // first claim size from the launch's events per warp
#endif
#ifndef LMOSEM_MIN_BATCH
#define LMOSEM_MIN_BATCH 4
#endif
#ifndef LMOSEM_GUIDED_LARGE
#define LMOSEM_GUIDED_LARGE 3  // guided divisor for launches of >= LMOSEM_GUIDED_ROUNDS rounds of claims
#endif
#ifndef LMOSEM_GUIDED_SMALL
#define LMOSEM_GUIDED_SMALL 2  // ... and for smaller ones (a rank's share at P >= 2); 0 = fixed claims
#endif
#ifndef LMOSEM_GUIDED_ROUNDS
#define LMOSEM_GUIDED_ROUNDS 6  // rounds = events / (32 x resident warps)
#endif
#ifndef LMOSEM_CLAIMS
#define LMOSEM_CLAIMS 4  // target claims per warp
#endif

// k_project work counters: {claimed events, exited warps} per slot, zeroed once at init;
// the last warp out of a launch re-zeroes its slot, so no memset precedes a launch
constexpr int kWorkSlots = 64;

// Path-buffer entries for a clip box whose largest extent is m voxels: <= 3 pieces per
// dominant-axis slab, >= 96 (the 32-event tile), rounded up to a multiple of 4 so every
// warp's buffer starts 32-byte aligned (the tile is staged with 16-byte vector stores).
int path_cap(int m) { return (std::max(96, 3 * m) + 3) & ~3; }

#ifndef LMOSEM_CAP_SUM
#define LMOSEM_CAP_SUM 1  // 0: size path buffers by 3 pieces per slab only (A/B)
#endif

// Path-buffer entries per warp for one launch: the forward-only modes (1, 2) keep no path
// and need only the 32-event tile (96 entries); the others hold the pieces of one LOR in the
// launch's clip box of extents e0, e1, e2 (the volume, or a slab of it). Two bounds: <= 3
// pieces per dominant-axis slab (3 max e), and one piece per slab plus one per minor-axis
// plane crossing: the minor positions stay inside the box up to rounding (lor_setup's guard),
// so each minor axis crosses at most e + 2 planes -> e_a + (e_b + 2) + (e_c + 2) <= sum e + 4.
// The smaller bound (C2: 584 instead of 840 pieces) leaves the SM more L1 for the gathers.
int launch_cap(int mode, const lmk::GridGeom& g) {
    if (mode == 1 || mode == 2) return 96;
    int m = 0, sum = 0;
    for (int k = 0; k < 3; ++k) {
        m = std::max(m, g.chi[k] - g.clo[k]);
        sum += g.chi[k] - g.clo[k];
    }
    if (LMOSEM_CAP_SUM && sum + 4 < 3 * m) return (std::max(96, sum + 4) + 3) & ~3;
    return path_cap(m);
}

// Resident CTAs per SM of k_project<mode> with `smem` bytes of path buffers (cached).
lmosem_status proj_occupancy(lmosem_ctx* ctx, int mode, size_t smem, int* blocks, bool list = false) {
    const int key = mode + (list ? 16 : 0);
    for (const auto& o : ctx->occ)
        if (o.mode == key && o.smem == smem) {
            *blocks = o.blocks;
            return LMOSEM_OK;
        }
    int b = 0;
    if (list) {
        switch (mode) {
            case 2: CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, lmk::k_project<2, true>, lmk::proj_threads_of(2), smem)); break;
            case 3: CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, lmk::k_project<3, true>, lmk::proj_threads_of(3), smem)); break;
            case 5: CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, lmk::k_project<5, true>, lmk::proj_threads_of(5), smem)); break;
            default: CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, lmk::k_project<6, true>, lmk::proj_threads_of(6), smem)); break;
        }
    } else switch (mode) {
        case 0: CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, lmk::k_project<0>, lmk::proj_threads_of(0), smem)); break;
        case 1: CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, lmk::k_project<1>, lmk::proj_threads_of(1), smem)); break;
        case 2: CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, lmk::k_project<2>, lmk::proj_threads_of(2), smem)); break;
        case 3: CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, lmk::k_project<3>, lmk::proj_threads_of(3), smem)); break;
        case 4: CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, lmk::k_project<4>, lmk::proj_threads_of(4), smem)); break;
        case 5: CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, lmk::k_project<5>, lmk::proj_threads_of(5), smem)); break;
        default: CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, lmk::k_project<6>, lmk::proj_threads_of(6), smem)); break;
    }
    b = std::max(1, b);
    ctx->occ.push_back({key, smem, b});
    *blocks = b;
    return LMOSEM_OK;
}

// la != nullptr (MODEs 2, 3, 5, 6): the launch runs over the listed events of *la (their
// number, <= n, is on the device; n sizes the grid)
lmosem_status launch_mode(lmosem_ctx* ctx, int mode, const float* evf, int64_t n, float* fp, const lmk::GridGeom& g,
                          const lmk::ListArg* la = nullptr) {
    const bool list = la != nullptr;
    const int cap = launch_cap(mode, g);
    const int threads = lmk::proj_threads_of(mode);
    const size_t sm = (threads / 32) * (sizeof(int2) * (size_t)cap + lmk::lor_bytes_per_warp(mode));
    int per_sm = 1;
    lmosem_status s = proj_occupancy(ctx, mode, sm, &per_sm, list);
    if (s) return s;
    const int64_t wpb = threads / 32;
    const int64_t resident = (int64_t)ctx->num_sms * per_sm * wpb;
    // events per claim: 32 when every warp gets >= 4 claims, else smaller (>= 4); the
    // kernel shrinks its claims further towards the end of the launch (guided)
    int batch = 32;
    while (LMOSEM_STATIC_BATCH && batch > LMOSEM_MIN_BATCH && n < (int64_t)batch * resident * LMOSEM_CLAIMS)
        batch >>= 1;
    const int64_t blocks_needed = ((n + batch - 1) / batch + wpb - 1) / wpb;
    const int64_t max_grid = (int64_t)ctx->num_sms * per_sm;
    const int grid = (int)std::max<int64_t>(1, std::min(blocks_needed, max_grid));
    unsigned long long* work = ctx->work + 2 * ctx->work_next;
    ctx->work_next = (ctx->work_next + 1) % kWorkSlots;
    // guided claims: a full C2/C5 subset (~9 rounds of 32-event claims per warp)
    // gains from the smaller final claims of divisor 3; a rank's share at P >= 2 from 2
    const int gdiv = n >= (int64_t)LMOSEM_GUIDED_ROUNDS * 32 * resident ? LMOSEM_GUIDED_LARGE : LMOSEM_GUIDED_SMALL;
    void (*k)(const float*, int64_t, const float*, float*, float*, lmk::GridGeom, int, unsigned long long*, int, int,
              lmk::ListArg);
    if (list) switch (mode) {
        case 2: k = lmk::k_project<2, true>; break;
        case 3: k = lmk::k_project<3, true>; break;
        case 5: k = lmk::k_project<5, true>; break;
        default: k = lmk::k_project<6, true>; break;
    } else switch (mode) {
        case 0: k = lmk::k_project<0>; break;
        case 1: k = lmk::k_project<1>; break;
        case 2: k = lmk::k_project<2>; break;
        case 3: k = lmk::k_project<3>; break;
        case 4: k = lmk::k_project<4>; break;
        case 5: k = lmk::k_project<5>; break;
        default: k = lmk::k_project<6>; break;
    }
    const lmk::ListArg none{};
    CK(launch_k(ctx, k, grid, threads, sm, evf, n, (const float*)ctx->fb, ctx->c, fp, g, cap, work, batch, gdiv,
                list ? *la : none));
    return LMOSEM_OK;
}

lmk::GridGeom slab_geom(const lmosem_ctx* ctx, int k, int K) {
    const int a = ctx->slab_axis;
    const int half = ctx->dims[a] / 2;  // slab boundaries on even coordinates (brick aligned)
    lmk::GridGeom g = ctx->geom;
    g.clo[a] = 2 * (int)((int64_t)half * k / K);
    g.chi[a] = (k == K - 1) ? ctx->dims[a] : 2 * (int)((int64_t)half * (k + 1) / K);
    return g;
}

// The listed z-slab form of step 1: k_zclass sorts the n events into
//   - the fine-window lists F_j (`wins`; LORs inside fine window j: one fused pass over the
//     window box, whose f and c fit L2 together),
//   - the medium-window lists M_j (`mwins`, coarse-slab wide; LORs inside one: passes A and B
//     over that window only),
//   - the coarse lists X_k (the other LORs: passes A and B over each coarse slab they meet).
// Order: pass A of every coarse slab k over [X_k, the M_j centred in slab k] (fp complete),
// then per coarse slab k one fused launch over the F_j centred in it and pass B over
// [X_k, M_j centred in it], so c's slab k stays L2-resident across them. The listed launches
// wait for their predecessor at exit (k_project, late_wait), except the first pass B.
lmosem_status launch_project_listed(lmosem_ctx* ctx, const float* evf, int64_t n, int K,
                                   const std::vector<std::pair<int, int>>& wins,
                                   const std::vector<std::pair<int, int>>& mwins) {
    const int Kf = (int)wins.size(), Km = (int)mwins.size();
    lmk::ZClass zc{};
    zc.K = K;
    zc.Kf = Kf;
    zc.Km = Km;
    zc.axis = ctx->slab_axis;
    for (int k = 0; k < K; ++k) {
        const lmk::GridGeom gk = slab_geom(ctx, k, K);
        zc.cb[k] = gk.clo[zc.axis];
        zc.cb[k + 1] = gk.chi[zc.axis];
    }
    for (int j = 0; j < Kf; ++j) {
        zc.wlo[j] = wins[j].first;
        zc.whi[j] = wins[j].second;
    }
    // a window family: starts j * stride (the last one clamped to end at the axis' end), equal widths
    auto family = [](const std::vector<std::pair<int, int>>& w, float& stride, float& width, float& last) {
        if (w.empty()) return;
        stride = w.size() > 1 ? (float)w[1].first : 1.0f;
        width = (float)(w[0].second - w[0].first);
        last = (float)w.back().first;
    };
    family(wins, zc.ws, zc.ww, zc.wlast);
    family(mwins, zc.ms, zc.mw, zc.mlast);
    not_kernel(ctx);
    CK(cudaMemsetAsync(ctx->zcount, 0, sizeof(int) * lmk::kZMaxLists, ctx->stream));
    CK(cudaMemsetAsync(ctx->fp_acc, 0, sizeof(float) * n, ctx->stream));
    const int zgrid = (int)std::max<int64_t>(1, std::min<int64_t>((n + lmk::kZChunk - 1) / lmk::kZChunk,
                                                                   (int64_t)ctx->num_sms * 8));
    CK(launch_k(ctx, lmk::k_zclass, zgrid, lmk::kZThreads, 0, evf, n, ctx->geom, zc, ctx->zlist, ctx->zlist_cap,
                ctx->zcount));
    // the first listed launch reads the lists before griddepcontrol.wait: a plain launch
    ctx->after_kernel = false;
    lmosem_status s;
    auto in_slab = [&](const std::pair<int, int>& w, int k) {  // a window runs with the slab of its centre
        const int mid = (w.first + w.second) / 2;
        return mid >= zc.cb[k] && mid < zc.cb[k + 1];
    };
    // passes A / B of region k: coarse slab k's list, then the medium windows centred in it
    // (each event clipped to its own segment's box; the path buffers sized for the widest)
    // k0..k1: the regions in one launch sequence (pass A of all regions may share launches)
    auto two_pass = [&](int mode, int k0, int k1) -> lmosem_status {
        struct Seg { int list, lo, hi; };
        std::vector<Seg> segs;
        for (int k = k0; k <= k1; ++k) {
            segs.push_back({k, zc.cb[k], zc.cb[k + 1]});
            for (int j = 0; j < Km; ++j)
                if (in_slab(mwins[j], k)) segs.push_back({K + Kf + j, mwins[j].first, mwins[j].second});
        }
        for (size_t i = 0; i < segs.size(); i += lmk::kMaxSeg) {
            lmk::ListArg la{};
            la.lists = ctx->zlist;
            la.counts = ctx->zcount;
            la.cap = ctx->zlist_cap;
            la.axis = zc.axis;
            la.box = 1;
            la.entry_wait = mode == 3 && k0 == 0 && i == 0;  // the first pass B waits for every pass A
            la.nseg = (int)std::min<size_t>(lmk::kMaxSeg, segs.size() - i);
            int widest = 0;
            for (int q = 0; q < la.nseg; ++q) {
                la.list[q] = segs[i + q].list;
                la.lo[q] = segs[i + q].lo;
                la.hi[q] = segs[i + q].hi;
                widest = std::max(widest, segs[i + q].hi - segs[i + q].lo);
            }
            lmk::GridGeom g = ctx->geom;  // only sizes the path buffers: the widest segment box
            g.clo[zc.axis] = 0;
            g.chi[zc.axis] = widest;
            if ((s = launch_mode(ctx, mode, evf, n, ctx->fp_acc, g, &la))) return s;
        }
        return LMOSEM_OK;
    };
    if (ctx->zamerge) {  // pass A of every region in as few launches as kMaxSeg allows
        if ((s = two_pass(2, 0, K - 1))) return s;
    } else {
        for (int k = 0; k < K; ++k)
            if ((s = two_pass(2, k, k))) return s;
    }
    const int fused = ctx->zfused_mode;
    for (int k = 0; k < K; ++k) {
        // the windows centred in slab k, in order, as one launch (up to kMaxSeg per launch, or
        // one per window with LMOSEM_ZMERGE=0): their lists are claimed in sequence, so the
        // LORs in flight stay within about one window
        int j = 0;
        while (j < Kf) {
            if (!in_slab(wins[j], k)) {
                ++j;
                continue;
            }
            lmk::ListArg la{};
            la.lists = ctx->zlist;
            la.counts = ctx->zcount;
            la.cap = ctx->zlist_cap;
            la.axis = zc.axis;
            la.box = 1;
            lmk::GridGeom gj = ctx->geom;  // the window box (equal widths: sizes the path buffers)
            gj.clo[zc.axis] = zc.wlo[j];
            gj.chi[zc.axis] = zc.whi[j];
            const int per = ctx->zmerge ? lmk::kMaxSeg : 1;
            for (; j < Kf && la.nseg < per && in_slab(wins[j], k); ++j) {
                la.list[la.nseg] = K + j;
                la.lo[la.nseg] = zc.wlo[j];
                la.hi[la.nseg] = zc.whi[j];
                la.nseg++;
            }
            if ((s = launch_mode(ctx, fused, evf, n, nullptr, gj, &la))) return s;
        }
        if ((s = two_pass(3, k, k))) return s;
    }
    return LMOSEM_OK;
}

// Step 1 over n device events against ctx->fb (mode 0: accumulate into ctx->c; mode 1:
// forward projections into fp_out; mode 4: sensitivity into ctx->c). Large images run
// the z-slab form (modes 0 -> 2 + 3; mode 4 slab by slab).
lmosem_status launch_project(lmosem_ctx* ctx, const lmosem_event* ev, int64_t n, float* fp_out, int mode) {
    if (n <= 0) return LMOSEM_OK;
    const float* evf = reinterpret_cast<const float*>(ev);
    const int K = n_slabs(ctx);
    if (mode == 1 || K == 1) {  // the fused pass gathers through the texture pipe when it can (MODE 5)
        int m = (mode == 0 && ctx->geom.tex_fb) ? 5 : mode;
        if (m == 5 && n >= ctx->wide_n) m = 6;  // large launch: 28 warps per SM
        return launch_mode(ctx, m, evf, n, fp_out, ctx->geom);
    }
    lmosem_status s;
    if (mode == 4) {
        for (int k = 0; k < K; ++k)
            if ((s = launch_mode(ctx, 4, evf, n, nullptr, slab_geom(ctx, k, K)))) return s;
        return LMOSEM_OK;
    }
    if (n > ctx->fp_cap) {
        if (ctx->fp_acc) CK(cudaFree(ctx->fp_acc));
        ctx->fp_acc = nullptr;
        ctx->fp_cap = 0;
        CKA(cudaMalloc(&ctx->fp_acc, sizeof(float) * n));
        ctx->fp_cap = n;
    }
    if (ctx->zlist_mode > 0 && n <= INT32_MAX && K <= lmk::kZMaxBits) {
        // fine windows along the slab axis (the fused launches gather through the texture
        // pipe, MODE 5/6): width ~ 1/zfine_per of a coarse slab, stride width/zover, even planes
        std::vector<std::pair<int, int>> wins, mwins;
        const int na = ctx->dims[ctx->slab_axis];
        // windows [l, l + width) every `stride` voxels (the last one ends at the axis' end)
        auto make = [na](std::vector<std::pair<int, int>>& w, int width, int stride) {
            w.clear();
            for (int lo = 0;; lo += stride) {
                const int l = std::min(lo, na - width);
                w.push_back({l, l + width});
                if (l + width >= na) break;
            }
        };
        const int W = ctx->zwin > 0 ? std::min(na, 2 * ((ctx->zwin + 1) / 2))
                                    : 2 * std::max(1, na / (2 * K * ctx->zfine_per));
        if (ctx->zlist_mode == 2 && ctx->geom.tex_fb && W < na) {
            // the stride grows (fewer, less overlapping windows) until the lists fit kZMaxLists
            for (int S = 2 * std::max(1, W / (2 * ctx->zover));; S += 2) {
                make(wins, W, S);
                if (K + (int)wins.size() <= lmk::kZMaxLists || S >= na) break;
            }
        }
        // medium windows (LMOSEM_ZMED > 0): as wide as a coarse slab, stride width / zmed, for
        // the LORs that leave every fine window but fit one coarse-slab width: passes A and B
        // over that one window instead of over each coarse slab they meet (with what is left
        // of the list budget; none if it does not fit)
        // default width 1.36 x the widest coarse slab (C4: 256 voxels, f or c of a window 95 MB;
        // measured 188 / 210 / 256 / 262 / 270 / 290 / 340: 21.31 / 21.33 / 20.93 / 20.96 /
        // 21.10 / 22.28 / 24.64 ms per subset, profiles/r02_zmwin_ab)
        const int Wm = ctx->zmwin > 0 ? std::min(na, 2 * ((ctx->zmwin + 1) / 2))
                                      : std::min(na, 2 * (int)(0.68 * max_slab_extent(na, K) + 0.5));
        if (ctx->zmed > 0 && K > 1 && Wm < na) {
            for (int S = 2 * std::max(1, Wm / (2 * ctx->zmed));; S += 2) {
                make(mwins, Wm, S);
                if (K + (int)wins.size() + (int)mwins.size() <= lmk::kZMaxLists || S >= na) break;  // >= 2 windows remain
            }
            if (K + (int)wins.size() + (int)mwins.size() > lmk::kZMaxLists) mwins.clear();
        }
        // the lists (allocated on first use, kept with the context); without the memory the
        // unlisted two-pass form runs instead
        const int nl = K + (int)wins.size() + (int)mwins.size();
        bool have = nl <= lmk::kZMaxLists && n <= ctx->zlist_cap && nl <= ctx->zlist_n && ctx->zcount;
        if (!have && nl <= lmk::kZMaxLists) {
            if (ctx->zlist) CK(cudaFree(ctx->zlist));
            ctx->zlist = nullptr;
            ctx->zlist_cap = 0;
            ctx->zlist_n = 0;
            if (cudaMalloc(&ctx->zlist, sizeof(int) * (size_t)n * nl) == cudaSuccess) {
                ctx->zlist_cap = n;
                ctx->zlist_n = nl;
            } else {
                (void)cudaGetLastError();  // out of memory is not sticky
                ctx->zlist = nullptr;
            }
            if (!ctx->zcount && cudaMalloc(&ctx->zcount, sizeof(int) * lmk::kZMaxLists) != cudaSuccess) {
                (void)cudaGetLastError();
                ctx->zcount = nullptr;
            }
            have = ctx->zlist && ctx->zcount;
        }
        if (have) return launch_project_listed(ctx, evf, n, K, wins, mwins);
    }
    not_kernel(ctx);
    CK(cudaMemsetAsync(ctx->fp_acc, 0, sizeof(float) * n, ctx->stream));
    for (int pass = 2; pass <= 3; ++pass)
        for (int k = 0; k < K; ++k)
            if ((s = launch_mode(ctx, pass, evf, n, ctx->fp_acc, slab_geom(ctx, k, K)))) return s;
    return LMOSEM_OK;
}

// step 2 on the bricks [b_begin, b_end); f_row (caller layout) is written when non-null;
// zero_to > 0 also re-zeroes c on every other brick of [0, zero_to) (ISD combine)
lmosem_status launch_update(lmosem_ctx* ctx, float* f_row, int64_t b_begin = 0, int64_t b_end = -1,
                            int64_t zero_to = 0) {
    if (b_end < 0) b_end = ctx->bricks.nb;
    const int64_t items = zero_to > 0 ? zero_to : b_end - b_begin;
    if (items <= 0) return LMOSEM_OK;
    CK(launch_k(ctx, lmk::k_update, grid_for(ctx, items), 256, 0, ctx->fb, ctx->c, (const float*)ctx->norm, f_row,
                ctx->geom, ctx->bricks, b_begin, b_end, zero_to));
    return LMOSEM_OK;
}

// NVTX range over one phase of a subset iteration (host enqueue side; nsys correlates the
// launches inside it). Costs a few ns without a tool attached.
struct Nvtx {
    explicit Nvtx(const char* name) { nvtxRangePushA(name); }
    void next(const char* name) {  // closes this range and opens the next phase's
        nvtxRangePop();
        nvtxRangePushA(name);
    }
    ~Nvtx() { nvtxRangePop(); }
};

// Destroying a failed context: abort the communicator so NCCL kernels stuck on a dead peer
// exit, and forget every handle tied to it.
void abort_comm(lmosem_ctx* ctx) {
    if (!ctx->comm) return;
    if (ctx->abort_flag) *(volatile int*)ctx->abort_flag = 1;
    ncclCommAbort(ctx->comm);
    ctx->comm = nullptr;
    ctx->dev_comm_ok = false;
    ctx->win_c = ctx->win_fb = nullptr;
    ctx->reg_c = ctx->reg_fb = nullptr;
}

// A collective failed or timed out: the context is failed (ENCCL, then ESTATE) and its
// communicator is aborted by lmosem_destroy (ncclCommAbort takes ~1 s of NCCL teardown, so
// the failing call returns first; the abort flag already stops the library's own kernels).
lmosem_status comm_failure(lmosem_ctx* ctx, lmosem_status s, const std::string& msg) {
    if (ctx->abort_flag) *(volatile int*)ctx->abort_flag = 1;
    return fail(ctx, s, msg);
}

// Waits until `ev` (or, with ev == nullptr, stream `st`) completes. With an NCCL
// communicator this is a watchdog: it polls ncclCommGetAsyncError and gives up after
// LMOSEM_TIMEOUT_S seconds (a peer that died or never joined the collective); the result is
// ENCCL, the context answers ESTATE from then on and lmosem_destroy aborts the communicator.
lmosem_status wait_done(lmosem_ctx* ctx, cudaStream_t st, cudaEvent_t ev = nullptr) {
    if (!ctx->comm) {
        CK(ev ? cudaEventSynchronize(ev) : cudaStreamSynchronize(st));
        return LMOSEM_OK;
    }
    const auto t0 = std::chrono::steady_clock::now();
    const double limit = coll_timeout_s();
    for (;;) {
        const cudaError_t e = ev ? cudaEventQuery(ev) : cudaStreamQuery(st);
        if (e == cudaSuccess) return LMOSEM_OK;
        if (e != cudaErrorNotReady)
            return comm_failure(ctx, LMOSEM_ECUDA, std::string("wait: ") + cudaGetErrorString(e));
        ncclResult_t ae = ncclSuccess;
        const ncclResult_t r = ncclCommGetAsyncError(ctx->comm, &ae);
        if (r != ncclSuccess || (ae != ncclSuccess && ae != ncclInProgress))
            return comm_failure(ctx, LMOSEM_ENCCL,
                                std::string("nccl async error: ") + ncclGetErrorString(r != ncclSuccess ? r : ae) +
                                    " (the communicator is aborted by lmosem_destroy)");
        const double waited = std::chrono::duration<double>(std::chrono::steady_clock::now() - t0).count();
        if (waited > limit)
            return comm_failure(ctx, LMOSEM_ENCCL,
                                "timed out after " + std::to_string((int)limit) +
                                    " s (LMOSEM_TIMEOUT_S) waiting for the stream: a peer rank stalled or died; the "
                                    "communicator is aborted by lmosem_destroy");
        std::this_thread::sleep_for(std::chrono::microseconds(50));
    }
}

lmosem_status mark(lmosem_ctx* ctx, PhaseMarks* pm, int k) {
    if (pm) {
        not_kernel(ctx);
        CK(cudaEventRecord(pm->e[k], ctx->stream));
    }
    return LMOSEM_OK;
}

lmosem_status get_marks(lmosem_ctx* ctx, PhaseMarks** out) {
    *out = nullptr;
    if (!ctx->timing) return LMOSEM_OK;
    if (ctx->pool.empty()) {
        PhaseMarks pm;
        for (int k = 0; k < 5; ++k) CK(cudaEventCreate(&pm.e[k]));
        ctx->pool.push_back(pm);
    }
    ctx->pending.push_back(ctx->pool.back());
    ctx->pool.pop_back();
    *out = &ctx->pending.back();
    return LMOSEM_OK;
}

// The final update can be split by brick z-planes (and f downloaded chunk by chunk) only
// when every rank updates its full replica (no ISD block split).
bool full_replica_update(const lmosem_ctx* ctx) {
    return !has_comm(ctx) || combine_mode(ctx) == LMOSEM_COMBINE_ALLREDUCE;
}

// Host-path pipelining of one subset iteration (reconstruct_host): in_chunks > 1 projects
// the events in in_chunks parts, part q after ev_pipe[q] (its upload) completed; host_f
// (with write_f, full_replica_update) runs the update in kPipe brick z-ranges and copies
// each finished range of f (device row layout) to host_f on the copy stream.
struct HostPipe {
    int in_chunks = 1;
    float* host_f = nullptr;
};

// One subset iteration on the context's stream: this rank's block of step 1, the c
// all-reduce (copy(add) -> every rank has the sum), step 2 on the full replica.
// to_brick: refresh ctx->fb from f first; write_f: write the updated f to the caller.
lmosem_status subset_iteration(lmosem_ctx* ctx, const lmosem_event* ev, int64_t n, float* f, bool whole_subset,
                               bool to_brick, bool write_f, const HostPipe& pipe = HostPipe()) {
    Nvtx range_subset("lmosem subset");
    int64_t b = 0, e = n;
    if (whole_subset) block_range(n, ctx->rank, ctx->world, &b, &e);
    PhaseMarks* pm = nullptr;
    lmosem_status s;
    if ((s = get_marks(ctx, &pm))) return s;
    if ((s = mark(ctx, pm, 0))) return s;
    if (to_brick && (s = launch_to_brick(ctx, f, ctx->fb))) return s;
    if ((s = mark(ctx, pm, 1))) return s;
    Nvtx range_project("lmosem project");  // then the combine + update
    if (pipe.in_chunks > 1) {
        for (int q = 0; q < pipe.in_chunks; ++q) {
            int64_t qb, qe;
            in_chunk_range(e - b, q, pipe.in_chunks, &qb, &qe);
            not_kernel(ctx);
            CK(cudaStreamWaitEvent(ctx->stream, ctx->ev_pipe[q], 0));
            if ((s = launch_project(ctx, ev + b + qb, qe - qb, nullptr, 0))) return s;
        }
    } else if ((s = launch_project(ctx, ev + b, e - b, nullptr, 0))) {
        return s;
    }
    if ((s = mark(ctx, pm, 2))) return s;
    range_project.next("lmosem combine + update");
    if (has_comm(ctx) && ctx->debug_stall_ms > 0) {  // tests of the watchdog only
        not_kernel(ctx);
        k_debug_stall<<<1, 32, 0, ctx->stream>>>(1000000ull * (unsigned long long)ctx->debug_stall_ms, ctx->abort_flag);
        CK(cudaGetLastError());
    }
    if (has_comm(ctx) && combine_mode(ctx) == LMOSEM_COMBINE_FUSED && (ctx->dev_comm_ok || ctx->loop)) {
        // NEXT-1: reduce-scatter + update + all-gather as one kernel over peer memory
        if ((s = coll_fused(ctx, ctx->nb_alloc / ctx->world))) return s;
        if ((s = mark(ctx, pm, 3))) return s;
        if (write_f && (s = launch_to_row(ctx, ctx->fb, f, 0))) return s;
    } else if (has_comm(ctx) && combine_mode(ctx) == LMOSEM_COMBINE_ISD) {
        // PAPER.md lines 509-518 (Listing 3 l.15-19): PSD -> ISD. Reduce-scatter c so rank r
        // holds the sum over its brick block, update only that block, all-gather f.
        const int64_t chunk = ctx->nb_alloc / ctx->world, b0 = chunk * ctx->rank;
        int64_t blk_b, blk_e, alloc;
        isd_block(ctx->bricks.nb, ctx->rank, ctx->world, &blk_b, &blk_e, &alloc);
        float* my_c = ctx->c + 8 * b0;
        if ((s = coll_reduce_scatter(ctx, ctx->c, my_c, (size_t)(8 * chunk)))) return s;
        // one launch: the block update (re-zeroes its c) and c <- 0 on every other brick
        if ((s = launch_update(ctx, nullptr, blk_b, blk_e, alloc))) return s;
        if ((s = coll_all_gather(ctx, ctx->fb + 8 * b0, ctx->fb, (size_t)(8 * chunk)))) return s;
        if ((s = mark(ctx, pm, 3))) return s;
        if (write_f && (s = launch_to_row(ctx, ctx->fb, f, 0))) return s;
    } else {
        if (has_comm(ctx) && (s = coll_all_reduce(ctx, ctx->c, (size_t)ctx->nbf))) return s;
        if ((s = mark(ctx, pm, 3))) return s;
        if (write_f && pipe.host_f) {
            // z-ranges of bricks: bricks [z0, z1) * BX*BY hold rows iz in [2 z0 - 2, 2 z1 - 2)
            const int64_t plane = (int64_t)ctx->bricks.BX * ctx->bricks.BY;
            const int64_t rowp = (int64_t)ctx->dims[0] * ctx->dims[1];
            for (int q = 0; q < kPipe; ++q) {
                int64_t z0, z1;
                block_range(ctx->bricks.BZ, q, kPipe, &z0, &z1);
                if ((s = launch_update(ctx, f, z0 * plane, z1 * plane))) return s;
                const int64_t r0 = std::max<int64_t>(0, 2 * z0 - lmk::HALO_LO);
                const int64_t r1 = std::min<int64_t>(ctx->dims[2], 2 * z1 - lmk::HALO_LO);
                if (r1 <= r0) continue;
                not_kernel(ctx);
                CK(cudaEventRecord(ctx->ev_pipe[q], ctx->stream));
                CK(cudaStreamWaitEvent(ctx->copy_stream, ctx->ev_pipe[q], 0));
                CK(cudaMemcpyAsync(pipe.host_f + r0 * rowp, f + r0 * rowp, sizeof(float) * (size_t)((r1 - r0) * rowp),
                                   cudaMemcpyDeviceToHost, ctx->copy_stream));
            }
        } else if ((s = launch_update(ctx, write_f ? f : nullptr))) {
            return s;
        }
    }
    if ((s = mark(ctx, pm, 4))) return s;
    ctx->st.subsets++;
    ctx->st.events += e - b;
    return LMOSEM_OK;
}

lmosem_status check_offsets(const int64_t* off, int32_t L) {
    if (!off || L < 0) return LMOSEM_EINVAL;
    if (off[0] < 0) return LMOSEM_EINVAL;
    for (int32_t l = 0; l < L; ++l)
        if (off[l + 1] < off[l]) return LMOSEM_EINVAL;
    return LMOSEM_OK;
}

lmosem_status resolve_timing(lmosem_ctx* ctx) {
    for (auto& pm : ctx->pending) {
        lmosem_status ws = wait_done(ctx, nullptr, pm.e[4]);
        if (ws) return ws;
        float t[4];
        for (int k = 0; k < 4; ++k) CK(cudaEventElapsedTime(&t[k], pm.e[k], pm.e[k + 1]));
        ctx->st.convert_ms += t[0];
        ctx->st.project_ms += t[1];
        ctx->st.combine_ms += t[2];
        ctx->st.update_ms += t[3];
        ctx->st.timed_subsets++;
        ctx->pool.push_back(pm);
    }
    ctx->pending.clear();
    for (size_t k = 0; k + 1 < ctx->h2d_pending.size(); k += 2) {
        lmosem_status ws = wait_done(ctx, nullptr, ctx->h2d_pending[k + 1]);
        if (ws) return ws;
        float t;
        CK(cudaEventElapsedTime(&t, ctx->h2d_pending[k], ctx->h2d_pending[k + 1]));
        ctx->st.h2d_ms += t;
        ctx->h2d_pool.push_back(ctx->h2d_pending[k]);
        ctx->h2d_pool.push_back(ctx->h2d_pending[k + 1]);
    }
    ctx->h2d_pending.clear();
    return LMOSEM_OK;
}

}  // namespace

#if LMK_TRACE
// diagnostic builds only (not declared in lmosem.h): the per-warp timeline of the last
// k_project launch (5 x uint64 per warp, see lmosem_kernels.cuh) to host memory, and reset
LMOSEM_API int lmosem_debug_trace(void* out, size_t bytes) {
    return cudaMemcpyFromSymbol(out, lmk::g_trace, std::min(bytes, sizeof(lmk::g_trace))) == cudaSuccess ? 0 : -1;
}
LMOSEM_API int lmosem_debug_trace_reset(void) {
    void* p = nullptr;
    if (cudaGetSymbolAddress(&p, lmk::g_trace) != cudaSuccess) return -1;
    return cudaMemset(p, 0, sizeof(lmk::g_trace)) == cudaSuccess ? 0 : -1;
}
#endif

LMOSEM_API const char* lmosem_version(void) { return "lmosem 0.5 sm_100a"; }

LMOSEM_API lmosem_status lmosem_block_range(int64_t n, int32_t rank, int32_t world, int64_t* begin, int64_t* end) {
    if (!begin || !end || n < 0 || world < 1 || rank < 0 || rank >= world) return LMOSEM_EINVAL;
    block_range(n, rank, world, begin, end);
    return LMOSEM_OK;
}

LMOSEM_API lmosem_status lmosem_isd_block(int64_t n_bricks, int32_t rank, int32_t world, int64_t* begin,
                                          int64_t* end, int64_t* alloc) {
    if (!begin || !end || !alloc || n_bricks < 0 || world < 1 || rank < 0 || rank >= world) return LMOSEM_EINVAL;
    isd_block(n_bricks, rank, world, begin, end, alloc);
    return LMOSEM_OK;
}

LMOSEM_API lmosem_status lmosem_nccl_unique_id(void* out, size_t size) {
    if (!out || size < sizeof(ncclUniqueId) || sizeof(ncclUniqueId) != LMOSEM_NCCL_ID_BYTES) return LMOSEM_EINVAL;
    ncclUniqueId id;
    if (ncclGetUniqueId(&id) != ncclSuccess) return LMOSEM_ENCCL;
    std::memcpy(out, &id, sizeof(id));
    return LMOSEM_OK;
}

namespace {

// A status with a message that leaves the context usable (unlike fail() for ENCCL/ECUDA).
lmosem_status soft_fail(lmosem_ctx* ctx, lmosem_status s, const std::string& msg) {
    ctx->err = msg;
    return s;
}

// Runs the fused combine once on the k_selftest_fill pattern (collective) and agrees on the
// verdict over the communicator (max of the mismatch counts); c and the brick f are zero
// again afterwards (f is refreshed from the caller's image at the next subset).
lmosem_status fused_selftest(lmosem_ctx* ctx, bool* passed) {
    *passed = false;
    const int64_t nbf_alloc = 8 * ctx->nb_alloc;
    float* ones = nullptr;
    int* bad = nullptr;
    CKA(cudaMalloc(&ones, sizeof(float) * nbf_alloc));
    if (cudaMalloc(&bad, sizeof(int)) != cudaSuccess) {
        cudaFree(ones);
        (void)cudaGetLastError();
        return fail(ctx, LMOSEM_ENOMEM, "fused self-test: cudaMalloc");
    }
    const float P = (float)ctx->world;
    lmosem_status s = LMOSEM_OK;
    float* norm = ctx->norm;
    ctx->norm = ones;  // the fused kernel reads the context's norm: s = 1 for the test
    int h_bad = -1;
    do {
        not_kernel(ctx);
        if (cudaMemsetAsync(bad, 0, sizeof(int), ctx->stream) != cudaSuccess) { s = fail(ctx, LMOSEM_ECUDA, "self-test memset"); break; }
        lmk::k_selftest_fill<<<grid_for(ctx, nbf_alloc), 256, 0, ctx->stream>>>(ctx->c, ctx->fb, ones, nbf_alloc,
                                                                                (float)(ctx->rank + 1));
        if ((s = coll_fused(ctx, ctx->nb_alloc / ctx->world))) break;
        lmk::k_selftest_check<<<grid_for(ctx, ctx->bricks.nb), 256, 0, ctx->stream>>>(ctx->c, ctx->fb, ctx->bricks,
                                                                                       0.5f * P * (P + 1.0f), bad);
        not_kernel(ctx);
        if (ncclAllReduce(bad, bad, 1, ncclInt32, ncclMax, ctx->comm, ctx->stream) != ncclSuccess) {
            s = fail(ctx, LMOSEM_ENCCL, "fused self-test: ncclAllReduce");
            break;
        }
        if (cudaMemcpyAsync(&h_bad, bad, sizeof(int), cudaMemcpyDeviceToHost, ctx->stream) != cudaSuccess ||
            cudaMemsetAsync(ctx->c, 0, sizeof(float) * nbf_alloc, ctx->stream) != cudaSuccess ||
            cudaMemsetAsync(ctx->fb, 0, sizeof(float) * nbf_alloc, ctx->stream) != cudaSuccess) {
            s = fail(ctx, LMOSEM_ECUDA, "fused self-test: copy");
            break;
        }
        s = wait_done(ctx, ctx->stream);
    } while (false);
    ctx->norm = norm;
    cudaFree(ones);
    cudaFree(bad);
    if (s) return s;
    *passed = h_bad == 0;
    return LMOSEM_OK;
}

// Collective set-up of the fused combine over NCCL: symmetric windows over c and the brick
// f, and a device communicator with one LSA barrier per CTA of the fused kernel (multimem
// when the team has it). On failure everything registered here is released again and the
// context stays usable (ENCCL with the reason in lmosem_last_error).
lmosem_status setup_fused(lmosem_ctx* ctx) {
    if (!ctx->comm || !ctx->nccl_mem)
        return soft_fail(ctx, LMOSEM_ENCCL, "set_combine(FUSED): needs a context with a dist and ncclMemAlloc images");
    CK(cudaStreamSynchronize(ctx->stream));
    const size_t bytes = sizeof(float) * 8 * ctx->nb_alloc;
    auto undo = [&](const std::string& why, ncclResult_t r) {
        if (ctx->win_c) ncclCommWindowDeregister(ctx->comm, ctx->win_c);
        if (ctx->win_fb) ncclCommWindowDeregister(ctx->comm, ctx->win_fb);
        ctx->win_c = ctx->win_fb = nullptr;
        return soft_fail(ctx, LMOSEM_ENCCL, "set_combine(FUSED): " + why + (r != ncclSuccess ? std::string(": ") + ncclGetErrorString(r) : ""));
    };
    ncclResult_t r = ncclCommWindowRegister(ctx->comm, ctx->c, bytes, &ctx->win_c, NCCL_WIN_COLL_SYMMETRIC);
    if (r != ncclSuccess) return (ctx->win_c = nullptr, undo("ncclCommWindowRegister(c)", r));
    r = ncclCommWindowRegister(ctx->comm, ctx->fb, bytes, &ctx->win_fb, NCCL_WIN_COLL_SYMMETRIC);
    if (r != ncclSuccess) return (ctx->win_fb = nullptr, undo("ncclCommWindowRegister(fb)", r));
    ctx->fused_ctas = LMOSEM_FUSED_CTAS_PER_SM * ctx->num_sms;  // all co-resident (barrier per CTA)
    ncclDevCommRequirements reqs;
    std::memset(&reqs, 0, sizeof(reqs));
    reqs.lsaBarrierCount = ctx->fused_ctas;
    reqs.lsaMultimem = ctx->world > 1;
    r = ncclDevCommCreate(ctx->comm, &reqs, &ctx->dev_comm);
    if (r != ncclSuccess && reqs.lsaMultimem) {
        reqs.lsaMultimem = false;
        r = ncclDevCommCreate(ctx->comm, &reqs, &ctx->dev_comm);
    }
    if (r != ncclSuccess) return undo("ncclDevCommCreate", r);
    if (ctx->dev_comm.lsaSize != ctx->world) {  // not one NVLink domain: keep the NCCL collectives
        ncclDevCommDestroy(ctx->comm, &ctx->dev_comm);
        return undo("the ranks are not one NVLink (LSA) domain", ncclSuccess);
    }
    ctx->dev_comm_ok = true;
    ctx->dev_comm_mm = reqs.lsaMultimem;
    bool passed = false;
    lmosem_status s = fused_selftest(ctx, &passed);
    if (s) return s;
    if (!passed) {
        ctx->dev_comm_ok = ctx->dev_comm_mm = false;
        ncclDevCommDestroy(ctx->comm, &ctx->dev_comm);
        return undo("self-test on the known pattern failed (kept the NCCL collectives)", ncclSuccess);
    }
    return LMOSEM_OK;
}

// Times the P > 1 combines on this box (collective; run at init after the fused combine's
// self-test): 2 warm-up and 5 timed runs each of the fused kernel, of reduce-scatter + block
// update + all-gather (ISD) and of all-reduce + full update, on the context's own images
// (zero at init, zero again after); the max over the ranks of each in ctx->st.tune_*_ms.
lmosem_status tune_combine(lmosem_ctx* ctx, bool with_fused) {
    const int64_t chunk = ctx->nb_alloc / ctx->world, b0 = chunk * ctx->rank;
    int64_t blk_b, blk_e, alloc;
    isd_block(ctx->bricks.nb, ctx->rank, ctx->world, &blk_b, &blk_e, &alloc);
    cudaEvent_t ev[2] = {nullptr, nullptr};
    float* d_t = nullptr;
    lmosem_status s = LMOSEM_OK;
    float t[3] = {0.f, 0.f, 0.f};
    auto run = [&](int which) -> lmosem_status {
        if (which == 0) return coll_fused(ctx, chunk);
        lmosem_status r;
        if (which == 2) {  // ALLREDUCE: all-reduce of c, then the full update on every rank
            if ((r = coll_all_reduce(ctx, ctx->c, (size_t)ctx->nbf))) return r;
            return launch_update(ctx, nullptr);
        }
        if ((r = coll_reduce_scatter(ctx, ctx->c, ctx->c + 8 * b0, (size_t)(8 * chunk)))) return r;
        if ((r = launch_update(ctx, nullptr, blk_b, blk_e, alloc))) return r;
        return coll_all_gather(ctx, ctx->fb + 8 * b0, ctx->fb, (size_t)(8 * chunk));
    };
    do {
        if (cudaEventCreate(&ev[0]) != cudaSuccess || cudaEventCreate(&ev[1]) != cudaSuccess ||
            cudaMalloc(&d_t, 3 * sizeof(float)) != cudaSuccess) {
            s = fail(ctx, LMOSEM_ECUDA, "tune_combine: events / buffer");
            break;
        }
        for (int which = with_fused ? 0 : 1; which < 3 && !s; ++which) {
            for (int i = 0; i < 2 && !s; ++i) s = run(which);
            if (s) break;
            not_kernel(ctx);
            if (cudaEventRecord(ev[0], ctx->stream) != cudaSuccess) {
                s = fail(ctx, LMOSEM_ECUDA, "tune_combine: record");
                break;
            }
            for (int i = 0; i < 5 && !s; ++i) s = run(which);
            if (s) break;
            not_kernel(ctx);
            if (cudaEventRecord(ev[1], ctx->stream) != cudaSuccess) {
                s = fail(ctx, LMOSEM_ECUDA, "tune_combine: record");
                break;
            }
            if ((s = wait_done(ctx, nullptr, ev[1]))) break;
            float ms = 0.f;
            cudaEventElapsedTime(&ms, ev[0], ev[1]);
            t[which] = ms / 5.f;
        }
        if (s) break;
        // agree on the times: max over the ranks
        not_kernel(ctx);
        if (cudaMemcpyAsync(d_t, t, sizeof(t), cudaMemcpyHostToDevice, ctx->stream) != cudaSuccess) {
            s = fail(ctx, LMOSEM_ECUDA, "tune_combine: copy");
            break;
        }
        if (ncclAllReduce(d_t, d_t, 3, ncclFloat32, ncclMax, ctx->comm, ctx->stream) != ncclSuccess) {
            s = fail(ctx, LMOSEM_ENCCL, "tune_combine: ncclAllReduce");
            break;
        }
        if (cudaMemcpyAsync(t, d_t, sizeof(t), cudaMemcpyDeviceToHost, ctx->stream) != cudaSuccess ||
            cudaMemsetAsync(ctx->c, 0, sizeof(float) * 8 * ctx->nb_alloc, ctx->stream) != cudaSuccess ||
            cudaMemsetAsync(ctx->fb, 0, sizeof(float) * 8 * ctx->nb_alloc, ctx->stream) != cudaSuccess) {
            s = fail(ctx, LMOSEM_ECUDA, "tune_combine: copy back");
            break;
        }
        s = wait_done(ctx, ctx->stream);
    } while (false);
    for (auto e : ev)
        if (e) cudaEventDestroy(e);
    if (d_t) cudaFree(d_t);
    if (s) return s;
    ctx->st.tune_fused_ms = t[0];
    ctx->st.tune_isd_ms = t[1];
    ctx->st.tune_allreduce_ms = t[2];
    return LMOSEM_OK;
}

}  // namespace

namespace {

// lmosem_init (dist: NCCL communicator) and lmosem_init_loopback (loop: loopback group)
lmosem_status init_ctx(lmosem_ctx** out, const int32_t dims[3], const double voxel_mm[3], const float* norm,
                       const lmosem_dist* dist, lmosem_loopback* loop, int32_t loop_rank) {
    if (!out) return LMOSEM_EINVAL;
    *out = nullptr;
    if (!dims || !voxel_mm || !norm) return LMOSEM_EINVAL;
    int64_t V = 1;
    for (int k = 0; k < 3; ++k) {
        if (dims[k] <= 0) return LMOSEM_EINVAL;
        if (!std::isfinite(voxel_mm[k]) || !(voxel_mm[k] > 0.0)) return LMOSEM_EINVAL;
        V *= dims[k];
    }
    if (V >= (int64_t(1) << 31)) return LMOSEM_EINVAL;
    // per-warp path buffer: 8 warps x 3 pieces per slab x 8 B must fit the 227 KB opt-in
    // shared memory of sm_100a for every clip box: one axis longer than kMaxBox is cut into
    // slabs (n_slabs), two are not supported (checked again against the device below)
    if ((dims[0] > kMaxBox) + (dims[1] > kMaxBox) + (dims[2] > kMaxBox) > 1) return LMOSEM_EINVAL;
    int rank = 0, world = 1;
    if (dist) {
        rank = dist->rank;
        world = dist->world;
        if (world < 1 || rank < 0 || rank >= world) return LMOSEM_EINVAL;
        if (!dist->nccl_unique_id) return LMOSEM_EINVAL;
    }
    if (loop) {
        rank = loop_rank;
        world = loop->world;
        if (rank < 0 || rank >= world) return LMOSEM_EINVAL;
    }
    lmosem_ctx* ctx = new (std::nothrow) lmosem_ctx;
    if (!ctx) return LMOSEM_ENOMEM;
    auto bail = [&](lmosem_status s) {
        g_init_err = ctx->err;
        lmosem_destroy(ctx);
        return s;
    };
    ctx->V = V;
    ctx->rank = rank;
    ctx->world = world;
    for (int k = 0; k < 3; ++k) {
        ctx->dims[k] = dims[k];
        ctx->vox[k] = voxel_mm[k];
        ctx->geom.n[k] = dims[k];
        ctx->geom.lo[k] = -0.5 * (double)dims[k] * voxel_mm[k];
        ctx->geom.v[k] = voxel_mm[k];
        ctx->geom.inv_v[k] = 1.0 / voxel_mm[k];
    }
    for (int k = 0; k < 3; ++k) {
        ctx->geom.clo[k] = 0;
        ctx->geom.chi[k] = dims[k];
    }
    // padded brick layout: halo of HALO_LO below, >= 2 above, even extents
    for (int k = 0; k < 3; ++k) ctx->geom.P[k] = (dims[k] + 4 + 1) & ~1;
    ctx->bricks.BX = ctx->geom.P[0] / 2;
    ctx->bricks.BY = ctx->geom.P[1] / 2;
    ctx->bricks.BZ = ctx->geom.P[2] / 2;
    ctx->bricks.nb = (int64_t)ctx->bricks.BX * ctx->bricks.BY * ctx->bricks.BZ;
    ctx->nbf = 8 * ctx->bricks.nb;
    for (int k = 0; k < 3; ++k) ctx->bricks.rhi[k] = (lmk::HALO_LO + dims[k] + 1) / 2;
    {
        int64_t b0, b1;
        isd_block(ctx->bricks.nb, rank, world, &b0, &b1, &ctx->nb_alloc);  // equal ISD brick blocks
    }
    if (ctx->nbf >= (int64_t(1) << 31)) {
        delete ctx;
        return LMOSEM_EINVAL;
    }
    {
        const int64_t M[3] = {8, 8LL * ctx->bricks.BX, 8LL * ctx->bricks.BX * ctx->bricks.BY};
        const int64_t m[3] = {1, 2, 4};
        for (int k = 0; k < 3; ++k) {
            ctx->geom.A[k] = (int)(M[k] / 2);
            ctx->geom.B[k] = (int)(m[k] - M[k] / 2);
        }
    }
    // slabs along z, or along the one axis longer than kMaxBox
    ctx->slab_axis = 2;
    for (int k = 0; k < 3; ++k)
        if (dims[k] > kMaxBox) ctx->slab_axis = k;
    // path buffer of the largest clip box (the whole volume, or a slab of it; see path_cap)
    {  // the largest clip box: the volume with its long axis clamped to kMaxBox (launch_cap's bounds)
        lmk::GridGeom box = ctx->geom;
        box.chi[ctx->slab_axis] = std::min(box.chi[ctx->slab_axis], kMaxBox);
        ctx->cap = launch_cap(0, box);
    }
    ctx->proj_smem = (lmk::PROJ_THREADS / 32) * (sizeof(int2) * (size_t)ctx->cap + lmk::lor_bytes_per_warp(0));

    lmosem_status s = LMOSEM_OK;
    auto cuda = [&](cudaError_t e, const char* what) {
        if (e != cudaSuccess && s == LMOSEM_OK) {
            s = (e == cudaErrorMemoryAllocation) ? LMOSEM_ENOMEM : LMOSEM_ECUDA;
            ctx->err = std::string(what) + ": " + cudaGetErrorString(e);
        }
        return e == cudaSuccess;
    };
    if (!cuda(cudaGetDevice(&ctx->device), "cudaGetDevice")) return bail(s);
    cudaDeviceProp prop;
    if (!cuda(cudaGetDeviceProperties(&prop, ctx->device), "cudaGetDeviceProperties")) return bail(s);
    ctx->num_sms = prop.multiProcessorCount;
    if (const char* e = std::getenv("LMOSEM_PDL")) ctx->pdl = e[0] != '0';  // A/B switch (default on)
    if (const char* e = std::getenv("LMOSEM_ZLIST")) ctx->zlist_mode = std::max(0, std::min(2, std::atoi(e)));
    if (const char* e = std::getenv("LMOSEM_ZFINE")) ctx->zfine_per = std::max(1, std::min(8, std::atoi(e)));
    if (const char* e = std::getenv("LMOSEM_ZFUSED_MODE")) ctx->zfused_mode = std::atoi(e) == 5 ? 5 : 6;
    if (const char* e = std::getenv("LMOSEM_ZOVER")) ctx->zover = std::max(1, std::min(4, std::atoi(e)));
    if (const char* e = std::getenv("LMOSEM_ZWIN")) ctx->zwin = std::max(0, std::atoi(e));
    if (const char* e = std::getenv("LMOSEM_ZMERGE")) ctx->zmerge = e[0] != '0';
    if (const char* e = std::getenv("LMOSEM_ZMED")) ctx->zmed = std::max(0, std::min(16, std::atoi(e)));
    if (const char* e = std::getenv("LMOSEM_ZAMERGE")) ctx->zamerge = e[0] != '0';
    if (const char* e = std::getenv("LMOSEM_ZMWIN")) ctx->zmwin = std::max(0, std::atoi(e));
    if (const char* e = std::getenv("LMOSEM_WIDE_N")) ctx->wide_n = std::max(0LL, std::atoll(e));
    if (const char* e = std::getenv("LMOSEM_DEBUG_STALL_MS")) ctx->debug_stall_ms = std::max(0, std::min(60000, std::atoi(e)));
    if (ctx->debug_stall_ms > 0) {
        if (!cuda(cudaHostAlloc(&ctx->abort_flag, sizeof(int), cudaHostAllocMapped), "cudaHostAlloc(abort flag)"))
            return bail(s);
        *ctx->abort_flag = 0;
    }
    if (ctx->proj_smem > (size_t)prop.sharedMemPerBlockOptin) {
        ctx->err = "volume too large for the shared-memory path buffer";
        return bail(LMOSEM_EINVAL);
    }


    // The limit is a per-function, process-wide attribute: set it to the device maximum
    // (not this context's need), so a smaller context created later cannot lower it under
    // a larger one (each launch passes its own size).
    {
        const int smax = (int)prop.sharedMemPerBlockOptin;
        // dynamic shared memory up to the opt-in limit less the kernel's static shared memory
        // (the listed variants keep their segment table there)
        auto smem_max = [&](auto kern) {
            cudaFuncAttributes fa{};
            cuda(cudaFuncGetAttributes(&fa, kern), "func attr");
            cuda(cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                      smax - (int)fa.sharedSizeBytes), "smem attr");
        };
        smem_max(lmk::k_project<0>);
        smem_max(lmk::k_project<1>);
        smem_max(lmk::k_project<2>);
        smem_max(lmk::k_project<3>);
        smem_max(lmk::k_project<4>);
        smem_max(lmk::k_project<5>);
        smem_max(lmk::k_project<6>);
        smem_max(lmk::k_project<2, true>);
        smem_max(lmk::k_project<3, true>);
        smem_max(lmk::k_project<5, true>);
        smem_max(lmk::k_project<6, true>);
    }
    cuda(cudaStreamCreateWithFlags(&ctx->own_stream, cudaStreamNonBlocking), "cudaStreamCreate");
    cuda(cudaStreamCreateWithFlags(&ctx->copy_stream, cudaStreamNonBlocking), "cudaStreamCreate");
    ctx->stream = ctx->own_stream;
    if (s != LMOSEM_OK) return bail(s);
    if (dist) {  // a communicator whenever a dist is given (world == 1 runs the 1-rank combine)
        ncclUniqueId id;
        std::memcpy(&id, dist->nccl_unique_id, sizeof(id));
        ncclResult_t r = ncclCommInitRank(&ctx->comm, world, id, rank);
        if (r != ncclSuccess) {
            ctx->comm = nullptr;
            ctx->err = std::string("ncclCommInitRank: ") + ncclGetErrorString(r);
            return bail(LMOSEM_ENCCL);
        }
        // the exchanged images come from ncclMemAlloc and are registered with the
        // communicator, so NCCL can run the reduce-scatter / all-gather zero-copy (and
        // through NVLS in-switch reduction on NVSwitch systems)
        const size_t bytes = sizeof(float) * 8 * ctx->nb_alloc;
        if (ncclMemAlloc((void**)&ctx->c, bytes) == ncclSuccess && ncclMemAlloc((void**)&ctx->fb, bytes) == ncclSuccess) {
            ctx->nccl_mem = true;
            if (ncclCommRegister(ctx->comm, ctx->c, bytes, &ctx->reg_c) != ncclSuccess) ctx->reg_c = nullptr;
            if (ncclCommRegister(ctx->comm, ctx->fb, bytes, &ctx->reg_fb) != ncclSuccess) ctx->reg_fb = nullptr;
        } else {
            if (ctx->c) ncclMemFree(ctx->c);
            if (ctx->fb) ncclMemFree(ctx->fb);
            ctx->c = ctx->fb = nullptr;
        }
    }
    if (!ctx->nccl_mem) {
        cuda(cudaMalloc(&ctx->c, sizeof(float) * 8 * ctx->nb_alloc), "cudaMalloc(c)");
        cuda(cudaMalloc(&ctx->fb, sizeof(float) * 8 * ctx->nb_alloc), "cudaMalloc(fb)");
    }
    cuda(cudaMalloc(&ctx->norm, sizeof(float) * 8 * ctx->nb_alloc), "cudaMalloc(norm)");
    cuda(cudaMalloc(&ctx->scratch, sizeof(float) * V), "cudaMalloc(scratch)");
    cuda(cudaMalloc(&ctx->work, sizeof(unsigned long long) * 2 * kWorkSlots), "cudaMalloc(work)");
    for (int k = 0; k < 2; ++k) {
        cuda(cudaEventCreateWithFlags(&ctx->ev_copied[k], cudaEventDisableTiming), "cudaEventCreate");
        cuda(cudaEventCreateWithFlags(&ctx->ev_consumed[k], cudaEventDisableTiming), "cudaEventCreate");
    }
    for (auto& e : ctx->ev_pipe) cuda(cudaEventCreateWithFlags(&e, cudaEventDisableTiming), "cudaEventCreate");
    if (loop)
        for (auto& e : ctx->loop_ev) cuda(cudaEventCreateWithFlags(&e, cudaEventDisableTiming), "cudaEventCreate");
    if (s != LMOSEM_OK) return bail(s);
    cuda(cudaMemcpyAsync(ctx->scratch, norm, sizeof(float) * V, cudaMemcpyDefault, ctx->stream), "copy norm");
    cuda(cudaMemsetAsync(ctx->c, 0, sizeof(float) * 8 * ctx->nb_alloc, ctx->stream), "memset c");
    cuda(cudaMemsetAsync(ctx->fb, 0, sizeof(float) * 8 * ctx->nb_alloc, ctx->stream), "memset fb");
    cuda(cudaMemsetAsync(ctx->norm, 0, sizeof(float) * 8 * ctx->nb_alloc, ctx->stream), "memset norm");
    cuda(cudaMemsetAsync(ctx->work, 0, sizeof(unsigned long long) * 2 * kWorkSlots, ctx->stream), "memset work");
    // MODE 5 (the fused pass with texture gathers) when the brick f fits a 1-D linear
    // texture; else, or with LMOSEM_TEX=0 (A/B, tests), the LSU gathers of MODE 0
    const char* te = std::getenv("LMOSEM_TEX");
    int max_lin = 0;
    cudaDeviceGetAttribute(&max_lin, cudaDevAttrMaxTexture1DLinearWidth, ctx->device);
    if (s == LMOSEM_OK && !(te && te[0] == '0') && 8 * ctx->nb_alloc <= (int64_t)max_lin) {
        cudaResourceDesc rd;
        std::memset(&rd, 0, sizeof(rd));
        rd.resType = cudaResourceTypeLinear;
        rd.res.linear.devPtr = ctx->fb;
        rd.res.linear.desc = cudaCreateChannelDesc<float>();
        rd.res.linear.sizeInBytes = sizeof(float) * 8 * ctx->nb_alloc;
        cudaTextureDesc td;
        std::memset(&td, 0, sizeof(td));
        td.readMode = cudaReadModeElementType;
        cudaTextureObject_t t = 0;
        if (cudaCreateTextureObject(&t, &rd, &td, nullptr) == cudaSuccess)
            ctx->geom.tex_fb = t;
        else
            (void)cudaGetLastError();  // not fatal: MODE 0 gathers
    }
    if (s == LMOSEM_OK) {
        lmk::k_row_to_brick<<<grid_for(ctx, ctx->bricks.nb), 256, 0, ctx->stream>>>(ctx->scratch, ctx->norm,
                                                                                     ctx->geom, ctx->bricks);
        cuda(cudaGetLastError(), "k_row_to_brick(norm)");
    }
    cuda(cudaStreamSynchronize(ctx->stream), "sync");
    if (s != LMOSEM_OK) return bail(s);
    // world > 1 over NCCL: set up the fused combine (NEXT-1) and self-test it (ISD, i.e.
    // reduce-scatter + all-gather, stays automatic when it fails or with LMOSEM_AUTO_FUSED=0).
    // If it sets up and passes, the three combines are timed on this box (tune_combine) and
    // the fastest becomes the automatic combine. LMOSEM_AUTO_FUSED=force does the same on a
    // 1-rank communicator (tests).
    {
        const char* af = std::getenv("LMOSEM_AUTO_FUSED");
        const bool force = af && std::strcmp(af, "force") == 0;
        if (ctx->comm && (world > 1 || force) && !(af && af[0] == '0')) {
            const lmosem_status fs = setup_fused(ctx);
            if (ctx->failed) return bail(fs);
            // without the fused combine (set-up or self-test failed) ISD and ALLREDUCE are timed
            const bool fused_ok = fs == LMOSEM_OK;
            const std::string why = ctx->err;
            const lmosem_status ts = tune_combine(ctx, fused_ok);
            if (ts) return bail(ts);
            ctx->err = why;
            const double tf = fused_ok ? ctx->st.tune_fused_ms : 1e30, ti = ctx->st.tune_isd_ms,
                         ta = ctx->st.tune_allreduce_ms;
            ctx->auto_combine = (tf <= ti && tf <= ta) ? LMOSEM_COMBINE_FUSED
                                                       : (ti <= ta ? LMOSEM_COMBINE_ISD : LMOSEM_COMBINE_ALLREDUCE);
        }
    }
    if (loop) {  // join the group: one context per rank, all on the group's device
        bool joined = false;
        {
            std::lock_guard<std::mutex> lk(loop->m);
            if (loop->device < 0) loop->device = ctx->device;
            if (loop->device == ctx->device && loop->ranks[rank] == nullptr) {
                loop->ranks[rank] = ctx;
                ctx->loop = loop;
                joined = true;
            }
        }
        if (!joined) {
            ctx->err = "init_loopback: rank already taken, or a different device than the group's";
            return bail(LMOSEM_EINVAL);
        }
    }
    *out = ctx;
    return LMOSEM_OK;
}

}  // namespace

LMOSEM_API lmosem_status lmosem_init(lmosem_ctx** out, const int32_t dims[3], const double voxel_mm[3],
                                     const float* norm, const lmosem_dist* dist) {
    return init_ctx(out, dims, voxel_mm, norm, dist, nullptr, 0);
}

LMOSEM_API lmosem_status lmosem_loopback_create(int32_t world, lmosem_loopback** out) {
    if (!out) return LMOSEM_EINVAL;
    *out = nullptr;
    if (world < 1 || world > lmk::kLoopMax) return LMOSEM_EINVAL;
    lmosem_loopback* g = new (std::nothrow) lmosem_loopback;
    if (!g) return LMOSEM_ENOMEM;
    g->world = world;
    g->ranks.assign(world, nullptr);
    g->src[0].assign(world, nullptr);
    g->src[1].assign(world, nullptr);
    *out = g;
    return LMOSEM_OK;
}

LMOSEM_API lmosem_status lmosem_loopback_destroy(lmosem_loopback* g) {
    if (!g) return LMOSEM_OK;
    {
        std::lock_guard<std::mutex> lk(g->m);
        for (auto* c : g->ranks)
            if (c) return LMOSEM_ESTATE;  // destroy the contexts first
    }
    if (g->bar) cudaFree(g->bar);
    delete g;
    return LMOSEM_OK;
}

LMOSEM_API lmosem_status lmosem_init_loopback(lmosem_ctx** out, const int32_t dims[3], const double voxel_mm[3],
                                              const float* norm, lmosem_loopback* group, int32_t rank) {
    if (!group) {
        if (out) *out = nullptr;
        return LMOSEM_EINVAL;
    }
    return init_ctx(out, dims, voxel_mm, norm, nullptr, group, rank);
}


LMOSEM_API lmosem_status lmosem_set_combine(lmosem_ctx* ctx, int32_t mode) {
    USABLE(ctx);
    if (mode < 0 || mode > LMOSEM_COMBINE_FUSED) return fail(ctx, LMOSEM_EINVAL, "set_combine: bad mode");
    if (mode == LMOSEM_COMBINE_FUSED && !ctx->dev_comm_ok && !ctx->loop) {
        lmosem_status s = setup_fused(ctx);
        if (s) return s;
    }
    ctx->combine = mode;
    return LMOSEM_OK;
}

LMOSEM_API int32_t lmosem_get_combine(const lmosem_ctx* ctx) { return ctx ? combine_mode(ctx) : -1; }

LMOSEM_API lmosem_status lmosem_set_slabs(lmosem_ctx* ctx, int32_t n_slabs) {
    USABLE(ctx);
    if (n_slabs < 0) return fail(ctx, LMOSEM_EINVAL, "set_slabs: n_slabs < 0");
    ctx->slabs_forced = n_slabs;
    return LMOSEM_OK;
}

LMOSEM_API int32_t lmosem_get_slabs(const lmosem_ctx* ctx) { return ctx ? n_slabs(ctx) : -1; }

LMOSEM_API lmosem_status lmosem_set_stream(lmosem_ctx* ctx, void* stream) {
    USABLE(ctx);
    ctx->stream = (cudaStream_t)stream;  // NULL = the CUDA default stream (e.g. torch's default)
    return LMOSEM_OK;
}

LMOSEM_API lmosem_status lmosem_subset_step(lmosem_ctx* ctx, const lmosem_event* events, int64_t n_events, float* f) {
    USABLE(ctx);
    if (!f || n_events < 0 || (n_events > 0 && !events)) return fail(ctx, LMOSEM_EINVAL, "subset_step: bad arguments");
    if (!device_accessible(f, n_events > 0 ? events : nullptr))
        return fail(ctx, LMOSEM_EINVAL, "subset_step: events / f are not device-accessible memory");
    if (events_misaligned(events, n_events)) return fail(ctx, LMOSEM_EINVAL, "subset_step: events not 8-byte aligned");
    return subset_iteration(ctx, events, n_events, f, true, true, true);
}

LMOSEM_API lmosem_status lmosem_reconstruct(lmosem_ctx* ctx, const lmosem_event* events, const int64_t* offsets,
                                            int32_t n_subsets, int32_t n_iterations, float* f) {
    USABLE(ctx);
    if (!f || n_iterations < 0 || check_offsets(offsets, n_subsets) || (offsets[n_subsets] > offsets[0] && !events))
        return fail(ctx, LMOSEM_EINVAL, "reconstruct: bad arguments");
    if (!device_accessible(f, offsets[n_subsets] > offsets[0] ? events : nullptr))
        return fail(ctx, LMOSEM_EINVAL, "reconstruct: events / f are not device-accessible memory");
    if (events_misaligned(events, offsets[n_subsets] - offsets[0]))
        return fail(ctx, LMOSEM_EINVAL, "reconstruct: events not 8-byte aligned");
    const int64_t total = (int64_t)n_iterations * n_subsets;
    int64_t step = 0;
    for (int32_t it = 0; it < n_iterations; ++it)
        for (int32_t l = 0; l < n_subsets; ++l, ++step) {
            lmosem_status s = subset_iteration(ctx, events + offsets[l], offsets[l + 1] - offsets[l], f, true,
                                               step == 0, step == total - 1);
            if (s) return s;
        }
    return LMOSEM_OK;
}

namespace {

// Device double buffers for streamed subsets (this rank's largest block).
lmosem_status ensure_stream_buffers(lmosem_ctx* ctx, const int64_t* offsets, int32_t n_subsets, bool pinned) {
    int64_t cap = 1;
    for (int32_t l = 0; l < n_subsets; ++l) {
        int64_t b, e;
        block_range(offsets[l + 1] - offsets[l], ctx->rank, ctx->world, &b, &e);
        cap = std::max(cap, e - b);
    }
    if (cap > ctx->dev_ev_cap) {
        for (int k = 0; k < 2; ++k) {
            if (ctx->dev_ev[k]) CK(cudaFree(ctx->dev_ev[k]));
            ctx->dev_ev[k] = nullptr;
        }
        ctx->dev_ev_cap = 0;
        for (int k = 0; k < 2; ++k) CKA(cudaMalloc(&ctx->dev_ev[k], sizeof(lmosem_event) * cap));
        ctx->dev_ev_cap = cap;
    }
    if (pinned && cap > ctx->pin_cap) {
        for (int k = 0; k < 2; ++k) {
            if (ctx->pin_ev[k]) CK(cudaFreeHost(ctx->pin_ev[k]));
            ctx->pin_ev[k] = nullptr;
        }
        ctx->pin_cap = 0;
        for (int k = 0; k < 2; ++k) CKA(cudaHostAlloc(&ctx->pin_ev[k], sizeof(lmosem_event) * cap, cudaHostAllocDefault));
        ctx->pin_cap = cap;
    }
    return LMOSEM_OK;
}

#ifndef LMOSEM_READ_THREADS
// reader threads of reconstruct_file; measured at C2 (16-core host, file in the page
// cache): 1/2/3/4/6/8/16 threads -> 3.7/6.0/7.7/8.3-8.7/8.2/7.3/7.3e8 events/s
#define LMOSEM_READ_THREADS 4
#endif

// Reads exactly `bytes` at `off` (retries short reads and EINTR).
bool pread_all(int fd, void* dst, size_t bytes, off_t off) {
    char* p = static_cast<char*>(dst);
    while (bytes > 0) {
        const ssize_t r = pread(fd, p, bytes, off);
        if (r < 0 && errno == EINTR) continue;
        if (r <= 0) return false;
        p += r;
        off += r;
        bytes -= (size_t)r;
    }
    return true;
}

// pread_all over up to LMOSEM_READ_THREADS threads in contiguous 1 MiB-aligned parts (page-cache reads are
// memcpy-bound per core; one thread reads ~8 GB/s, a 24 MB subset block then takes longer
// than its projection).
bool pread_parallel(int fd, void* dst, size_t bytes, off_t off) {
    const size_t min_part = size_t(1) << 20;
    const unsigned hw = std::max(1u, std::thread::hardware_concurrency());
    const size_t nt = std::min<size_t>(std::min<size_t>(LMOSEM_READ_THREADS, hw), std::max<size_t>(1, bytes / min_part));
    if (nt <= 1) return pread_all(fd, dst, bytes, off);
    std::vector<std::thread> th;
    std::vector<char> ok(nt, 1);
    const size_t part = (bytes / nt + 4095) & ~size_t(4095);
    for (size_t t = 0; t < nt; ++t) {
        const size_t b = std::min(bytes, t * part), e = std::min(bytes, (t + 1) * part);
        if (e <= b) break;
        th.emplace_back([&, t, b, e] { ok[t] = pread_all(fd, static_cast<char*>(dst) + b, e - b, off + (off_t)b); });
    }
    for (auto& x : th) x.join();
    for (char o : ok)
        if (!o) return false;
    return true;
}

}  // namespace

LMOSEM_API lmosem_status lmosem_reconstruct_file(lmosem_ctx* ctx, const char* path, const int64_t* offsets,
                                                 int32_t n_subsets, int32_t n_iterations, float* f) {
    USABLE(ctx);
    if (!path || !f || n_iterations < 0 || check_offsets(offsets, n_subsets))
        return fail(ctx, LMOSEM_EINVAL, "reconstruct_file: bad arguments");
    if (!device_accessible(f)) return fail(ctx, LMOSEM_EINVAL, "reconstruct_file: f is not device-accessible memory");
    const int fd = open(path, O_RDONLY);
    if (fd < 0) return fail(ctx, LMOSEM_EIO, std::string("reconstruct_file: open ") + path + ": " + strerror(errno));
    struct stat sb;
    if (fstat(fd, &sb) != 0 || (int64_t)sb.st_size < offsets[n_subsets] * (int64_t)sizeof(lmosem_event)) {
        close(fd);
        return fail(ctx, LMOSEM_EIO, std::string("reconstruct_file: ") + path + " is shorter than offsets[n_subsets]");
    }
    lmosem_status s = ensure_stream_buffers(ctx, offsets, n_subsets, true);
    if (s) {
        close(fd);
        return s;
    }
    // staging buffer k is free once the H2D copy out of it (ev_copied[k]) completed;
    // device buffer k is free once the projection of its subset (ev_consumed[k]) completed
    for (int k = 0; k < 2; ++k) {
        if (cudaEventRecord(ctx->ev_consumed[k], ctx->stream) != cudaSuccess ||
            cudaEventRecord(ctx->ev_copied[k], ctx->copy_stream) != cudaSuccess) {
            close(fd);
            return fail(ctx, LMOSEM_ECUDA, "reconstruct_file: cudaEventRecord");
        }
    }
    int64_t step = 0;
    const int64_t total = (int64_t)n_iterations * n_subsets;
    for (int32_t it = 0; it < n_iterations && !s; ++it)
        for (int32_t l = 0; l < n_subsets && !s; ++l, ++step) {
            const int k = (int)(step & 1);
            int64_t b, e;
            block_range(offsets[l + 1] - offsets[l], ctx->rank, ctx->world, &b, &e);
            // host: read this rank's block while the GPU works on the previous subset
            if ((s = wait_done(ctx, nullptr, ctx->ev_copied[k]))) break;
            if (e > b && !pread_parallel(fd, ctx->pin_ev[k], sizeof(lmosem_event) * (e - b),
                                         (off_t)(sizeof(lmosem_event) * (offsets[l] + b)))) {
                s = fail(ctx, LMOSEM_EIO, std::string("reconstruct_file: read ") + path + ": " + strerror(errno));
                break;
            }
            not_kernel(ctx);  // the wait on ctx->stream below
            if (cudaStreamWaitEvent(ctx->copy_stream, ctx->ev_consumed[k], 0) != cudaSuccess ||
                (e > b && cudaMemcpyAsync(ctx->dev_ev[k], ctx->pin_ev[k], sizeof(lmosem_event) * (e - b),
                                          cudaMemcpyHostToDevice, ctx->copy_stream) != cudaSuccess) ||
                cudaEventRecord(ctx->ev_copied[k], ctx->copy_stream) != cudaSuccess ||
                cudaStreamWaitEvent(ctx->stream, ctx->ev_copied[k], 0) != cudaSuccess) {
                s = fail(ctx, LMOSEM_ECUDA, "reconstruct_file: upload");
                break;
            }
            s = subset_iteration(ctx, ctx->dev_ev[k], e - b, f, false, step == 0, step == total - 1);
            if (!s && cudaEventRecord(ctx->ev_consumed[k], ctx->stream) != cudaSuccess)
                s = fail(ctx, LMOSEM_ECUDA, "reconstruct_file: cudaEventRecord");
        }
    close(fd);
    if (s == LMOSEM_EIO) {  // nothing left in flight on return
        const std::string msg = ctx->err;
        lmosem_status ws = wait_done(ctx, ctx->stream);
        if (ws) return ws;
        ctx->err = msg;
    }
    if (s) return s;
    return wait_done(ctx, ctx->stream);
}

LMOSEM_API lmosem_status lmosem_reconstruct_host(lmosem_ctx* ctx, const lmosem_event* events, const int64_t* offsets,
                                                 int32_t n_subsets, int32_t n_iterations, float* f) {
    USABLE(ctx);
    if (!f || n_iterations < 0 || check_offsets(offsets, n_subsets) || (offsets[n_subsets] > offsets[0] && !events))
        return fail(ctx, LMOSEM_EINVAL, "reconstruct_host: bad arguments");
    // this rank's block of every subset: the only events it uploads (block distribution)
    lmosem_status s0 = ensure_stream_buffers(ctx, offsets, n_subsets, false);
    if (s0) return s0;
    if (!ctx->dev_f) CKA(cudaMalloc(&ctx->dev_f, sizeof(float) * ctx->V));
    // f goes up first on the copy stream (the first projection needs it), then the first
    // subset's events in kPipe chunks that the projection consumes as they land
    CK(cudaEventRecord(ctx->ev_pipe[kPipe], ctx->stream));
    CK(cudaStreamWaitEvent(ctx->copy_stream, ctx->ev_pipe[kPipe], 0));
    CK(cudaMemcpyAsync(ctx->dev_f, f, sizeof(float) * ctx->V, cudaMemcpyHostToDevice, ctx->copy_stream));
    CK(cudaEventRecord(ctx->ev_pipe[kPipe], ctx->copy_stream));
    CK(cudaStreamWaitEvent(ctx->stream, ctx->ev_pipe[kPipe], 0));
    // buffers start free
    for (int k = 0; k < 2; ++k) CK(cudaEventRecord(ctx->ev_consumed[k], ctx->stream));
    int64_t step = 0;
    const int64_t total = (int64_t)n_iterations * n_subsets;
    const bool pipe_out = full_replica_update(ctx);
    for (int32_t it = 0; it < n_iterations; ++it)
        for (int32_t l = 0; l < n_subsets; ++l, ++step) {
            const int k = (int)(step & 1);
            int64_t b, e;
            block_range(offsets[l + 1] - offsets[l], ctx->rank, ctx->world, &b, &e);
            not_kernel(ctx);  // the event record / wait on ctx->stream around this subset
            CK(cudaStreamWaitEvent(ctx->copy_stream, ctx->ev_consumed[k], 0));
            cudaEvent_t h0 = nullptr, h1 = nullptr;
            if (ctx->timing) {
                for (int q = 0; q < 2; ++q) {
                    if (ctx->h2d_pool.empty()) {
                        cudaEvent_t ev;
                        CK(cudaEventCreate(&ev));
                        ctx->h2d_pool.push_back(ev);
                    }
                    (q ? h1 : h0) = ctx->h2d_pool.back();
                    ctx->h2d_pool.pop_back();
                }
                CK(cudaEventRecord(h0, ctx->copy_stream));
            }
            HostPipe pipe;
            // nothing to overlap the first subset's upload with: chunk it (>= 64 K events per chunk)
            if (step == 0 && e - b >= (int64_t)16 * 16384) pipe.in_chunks = kInChunks;
            for (int q = 0; q < pipe.in_chunks; ++q) {
                int64_t qb, qe;
                in_chunk_range(e - b, q, pipe.in_chunks, &qb, &qe);
                if (qe > qb)
                    CK(cudaMemcpyAsync(ctx->dev_ev[k] + qb, events + offsets[l] + b + qb, sizeof(lmosem_event) * (qe - qb),
                                       cudaMemcpyHostToDevice, ctx->copy_stream));
                if (pipe.in_chunks > 1) CK(cudaEventRecord(ctx->ev_pipe[q], ctx->copy_stream));
            }
            if (ctx->timing) {
                CK(cudaEventRecord(h1, ctx->copy_stream));
                ctx->h2d_pending.push_back(h0);
                ctx->h2d_pending.push_back(h1);
            }
            CK(cudaEventRecord(ctx->ev_copied[k], ctx->copy_stream));
            if (pipe.in_chunks == 1) CK(cudaStreamWaitEvent(ctx->stream, ctx->ev_copied[k], 0));
            if (pipe_out && step == total - 1) pipe.host_f = f;
            lmosem_status s = subset_iteration(ctx, ctx->dev_ev[k], e - b, ctx->dev_f, false, step == 0,
                                               step == total - 1, pipe);
            if (s) return s;
            CK(cudaEventRecord(ctx->ev_consumed[k], ctx->stream));
        }
    if (!pipe_out || total == 0)
        CK(cudaMemcpyAsync(f, ctx->dev_f, sizeof(float) * ctx->V, cudaMemcpyDeviceToHost, ctx->stream));
    lmosem_status ws = wait_done(ctx, ctx->stream);
    if (ws) return ws;
    return wait_done(ctx, ctx->copy_stream);
}

LMOSEM_API lmosem_status lmosem_error_image(lmosem_ctx* ctx, const lmosem_event* events, int64_t n_events,
                                            const float* f, float* c_out) {
    USABLE(ctx);
    if (!f || !c_out || n_events < 0 || (n_events > 0 && !events))
        return fail(ctx, LMOSEM_EINVAL, "error_image: bad arguments");
    if (!device_accessible(f, c_out, n_events > 0 ? events : nullptr))
        return fail(ctx, LMOSEM_EINVAL, "error_image: buffers are not device-accessible memory");
    if (events_misaligned(events, n_events)) return fail(ctx, LMOSEM_EINVAL, "error_image: events not 8-byte aligned");
    lmosem_status s;
    if ((s = launch_to_brick(ctx, f, ctx->fb))) return s;
    if ((s = launch_project(ctx, events, n_events, nullptr, 0))) return s;
    return launch_to_row(ctx, ctx->c, c_out, 1);  // c_out <- c, c <- 0
}

LMOSEM_API lmosem_status lmosem_forward(lmosem_ctx* ctx, const lmosem_event* events, int64_t n_events,
                                        const float* f, float* fp_out) {
    USABLE(ctx);
    if (!f || n_events < 0 || (n_events > 0 && (!events || !fp_out)))
        return fail(ctx, LMOSEM_EINVAL, "forward: bad arguments");
    if (!device_accessible(f, n_events > 0 ? events : nullptr, n_events > 0 ? fp_out : nullptr))
        return fail(ctx, LMOSEM_EINVAL, "forward: buffers are not device-accessible memory");
    if (events_misaligned(events, n_events)) return fail(ctx, LMOSEM_EINVAL, "forward: events not 8-byte aligned");
    lmosem_status s;
    if ((s = launch_to_brick(ctx, f, ctx->fb))) return s;
    return launch_project(ctx, events, n_events, fp_out, 1);
}

LMOSEM_API lmosem_status lmosem_sensitivity(lmosem_ctx* ctx, const lmosem_event* events, int64_t n_events,
                                            float* s_out) {
    USABLE(ctx);
    if (!s_out || n_events < 0 || (n_events > 0 && !events))
        return fail(ctx, LMOSEM_EINVAL, "sensitivity: bad arguments");
    if (!device_accessible(s_out, n_events > 0 ? events : nullptr))
        return fail(ctx, LMOSEM_EINVAL, "sensitivity: buffers are not device-accessible memory");
    if (events_misaligned(events, n_events)) return fail(ctx, LMOSEM_EINVAL, "sensitivity: events not 8-byte aligned");
    int64_t b = 0, e = n_events;
    block_range(n_events, ctx->rank, ctx->world, &b, &e);
    lmosem_status s;
    if ((s = launch_project(ctx, events + b, e - b, nullptr, 4))) return s;
    if (has_comm(ctx) && (s = coll_all_reduce(ctx, ctx->c, (size_t)ctx->nbf))) return s;
    return launch_to_row(ctx, ctx->c, s_out, 1);  // s_out <- c, c <- 0
}

LMOSEM_API lmosem_status lmosem_set_norm(lmosem_ctx* ctx, const float* norm) {
    USABLE(ctx);
    if (!norm) return fail(ctx, LMOSEM_EINVAL, "set_norm: null norm");
    CK(cudaMemcpyAsync(ctx->scratch, norm, sizeof(float) * ctx->V, cudaMemcpyDefault, ctx->stream));
    lmosem_status s = launch_to_brick(ctx, ctx->scratch, ctx->norm);
    if (s) return s;
    return wait_done(ctx, ctx->stream);  // the caller may release `norm` on return
}

LMOSEM_API lmosem_status lmosem_update(lmosem_ctx* ctx, float* f, float* c) {
    USABLE(ctx);
    if (!f || !c) return fail(ctx, LMOSEM_EINVAL, "update: bad arguments");
    if (!device_accessible(f, c)) return fail(ctx, LMOSEM_EINVAL, "update: f / c are not device-accessible memory");
    lmosem_status s;
    if ((s = launch_to_brick(ctx, f, ctx->fb))) return s;
    if ((s = launch_to_brick(ctx, c, ctx->c))) return s;
    if ((s = launch_update(ctx, f))) return s;  // also re-zeroes the context's c
    CK(cudaMemsetAsync(c, 0, sizeof(float) * ctx->V, ctx->stream));
    return LMOSEM_OK;
}

LMOSEM_API lmosem_status lmosem_synchronize(lmosem_ctx* ctx) {
    USABLE(ctx);
    lmosem_status s = wait_done(ctx, ctx->stream);
    if (s) return s;
    if ((s = wait_done(ctx, ctx->copy_stream))) return s;
    if (ctx->comm) {
        ncclResult_t async_err = ncclSuccess;
        NK(ncclCommGetAsyncError(ctx->comm, &async_err));
        if (async_err != ncclSuccess)
            return comm_failure(ctx, LMOSEM_ENCCL, std::string("nccl async: ") + ncclGetErrorString(async_err));
    }
    return LMOSEM_OK;
}

LMOSEM_API lmosem_status lmosem_set_timing(lmosem_ctx* ctx, int32_t enable) {
    USABLE(ctx);
    lmosem_status s = resolve_timing(ctx);
    if (s) return s;
    ctx->timing = enable != 0;
    if (ctx->timing) {
        ctx->st.convert_ms = ctx->st.project_ms = ctx->st.combine_ms = ctx->st.update_ms = ctx->st.h2d_ms = 0.0;
        ctx->st.timed_subsets = 0;
    }
    return LMOSEM_OK;
}

LMOSEM_API lmosem_status lmosem_get_stats(lmosem_ctx* ctx, lmosem_stats* out) {
    USABLE(ctx);
    if (!out) return LMOSEM_EINVAL;
    lmosem_status s = resolve_timing(ctx);
    if (s) return s;
    *out = ctx->st;
    return LMOSEM_OK;
}

LMOSEM_API lmosem_status lmosem_destroy(lmosem_ctx* ctx) {
    if (!ctx) return LMOSEM_OK;
    // a failed context may have a collective stuck on a dead peer: abort the communicator
    // before waiting for the streams (its kernels then exit)
    if (ctx->failed) abort_comm(ctx);
    if (ctx->stream) cudaStreamSynchronize(ctx->stream);
    if (ctx->copy_stream) cudaStreamSynchronize(ctx->copy_stream);
    if (ctx->comm) {
        if (ctx->dev_comm_ok) ncclDevCommDestroy(ctx->comm, &ctx->dev_comm);
        if (ctx->win_c) ncclCommWindowDeregister(ctx->comm, ctx->win_c);
        if (ctx->win_fb) ncclCommWindowDeregister(ctx->comm, ctx->win_fb);
        if (ctx->reg_c) ncclCommDeregister(ctx->comm, ctx->reg_c);
        if (ctx->reg_fb) ncclCommDeregister(ctx->comm, ctx->reg_fb);
    }
    if (ctx->nccl_mem) {
        if (ctx->c) ncclMemFree(ctx->c);
        if (ctx->fb) ncclMemFree(ctx->fb);
        ctx->c = ctx->fb = nullptr;
    }
    if (ctx->comm) ncclCommDestroy(ctx->comm);
    if (ctx->loop) {
        std::lock_guard<std::mutex> lk(ctx->loop->m);
        ctx->loop->ranks[ctx->rank] = nullptr;
    }
    for (auto e : ctx->loop_ev)
        if (e) cudaEventDestroy(e);
    for (auto& pm : ctx->pending)
        for (int k = 0; k < 5; ++k) cudaEventDestroy(pm.e[k]);
    for (auto& pm : ctx->pool)
        for (int k = 0; k < 5; ++k) cudaEventDestroy(pm.e[k]);
    for (auto e : ctx->h2d_pending) cudaEventDestroy(e);
    for (auto e : ctx->h2d_pool) cudaEventDestroy(e);
    for (int k = 0; k < 2; ++k) {
        if (ctx->pin_ev[k]) cudaFreeHost(ctx->pin_ev[k]);
        if (ctx->dev_ev[k]) cudaFree(ctx->dev_ev[k]);
        if (ctx->ev_copied[k]) cudaEventDestroy(ctx->ev_copied[k]);
        if (ctx->ev_consumed[k]) cudaEventDestroy(ctx->ev_consumed[k]);
    }
    for (auto e : ctx->ev_pipe)
        if (e) cudaEventDestroy(e);
    if (ctx->dev_f) cudaFree(ctx->dev_f);
    if (ctx->abort_flag) cudaFreeHost(ctx->abort_flag);
    if (ctx->geom.tex_fb) cudaDestroyTextureObject(ctx->geom.tex_fb);
    if (ctx->c) cudaFree(ctx->c);
    if (ctx->fb) cudaFree(ctx->fb);
    if (ctx->norm) cudaFree(ctx->norm);
    if (ctx->scratch) cudaFree(ctx->scratch);
    if (ctx->fp_acc) cudaFree(ctx->fp_acc);
    if (ctx->zlist) cudaFree(ctx->zlist);
    if (ctx->zcount) cudaFree(ctx->zcount);
    if (ctx->work) cudaFree(ctx->work);
    if (ctx->own_stream) cudaStreamDestroy(ctx->own_stream);
    if (ctx->copy_stream) cudaStreamDestroy(ctx->copy_stream);
    delete ctx;
    return LMOSEM_OK;
}

LMOSEM_API const char* lmosem_last_error(const lmosem_ctx* ctx) {
    if (!ctx) return g_init_err.empty() ? "lmosem: null context" : g_init_err.c_str();
    return ctx->err.c_str();
}
