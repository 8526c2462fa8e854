/* lmosem.h — C ABI of the B200-native LM-OSEM subset iteration.
 *
 * The operation (§IV, Listing 2; Listing 3):
 * list-mode OSEM reconstructs an image f from events (lines of response, LORs) split
 * into subsets. One subset iteration is
 *   step 1 (Listing 2 lines 5-13): c <- 0; for every event i of the subset,
 *            path_i = compute_path(event_i)                   exact Siddon chord lengths a_ij
 *            fp_i   = sum_j a_ij f_j                          forward projection
 *            c_j   += a_ij / fp_i  for j on path_i            back-projection (skip fp_i <= 0)
 *   combine (Listing 3 lines 6, 15-16): with several GPUs the
 *            per-GPU error images are added element-wise (copy(add) distribution)
 *   step 2 (Listing 2 lines 16-17 with the norm of BASELINE.json north_star):
 *            f_j <- f_j * c_j / s_j  where c_j > 0 and s_j > 0, else unchanged.
 * Readings of points the paper leaves open are listed in DESIGN.md (S1-S17).
 *
 * Conventions
 *  - Volume: nx*ny*nz voxels of vx*vy*vz mm, centred on the origin. Voxel (ix,iy,iz) is
 *    the half-open box [x0+ix*vx, x0+(ix+1)*vx) x ..., x0 = -nx*vx/2; images are float32
 *    with linear index j = ix + nx*(iy + ny*iz) (x fastest). V = nx*ny*nz < 2^31.
 *  - Event: lmosem_event, 6 float32 (two detection points in mm, the segment p1 -> p2).
 *    Device event arrays must be 8-byte aligned (EINVAL otherwise).
 *    Non-finite, zero-length or volume-missing events, and events with fp_i <= 0,
 *    contribute nothing (not an error).
 *  - Pointers: "device" = CUDA device memory of the context's device; "host" = host
 *    memory (pinned memory gives overlapped copies). The caller owns every buffer it
 *    passes; the context owns c, its copy of the norm image, scratch buffers, its
 *    streams and (world > 1) its NCCL communicator.
 *  - Ordering: calls taking device buffers are enqueued on the context's stream (see
 *    lmosem_set_stream) and return without waiting; lmosem_synchronize waits. Calls
 *    taking host buffers are synchronous.
 *  - Distribution (§III.A; §IV.A): with
 *    world > 1, subset_step / reconstruct are collective. Every rank passes the WHOLE
 *    subset; rank r projects the block [floor(r*N/P), floor((r+1)*N/P)) (block
 *    distribution), f is replicated (copy distribution) and c is combined over NVLink
 *    (copy(add)) by the paper's PSD -> ISD switch — reduce-scatter, block update,
 *    all-gather — as one fused multimem kernel when available (else NCCL collectives), or
 *    by an all-reduce + full update (lmosem_set_combine). Either way the replicas of f are
 *    identical on return. A loopback group (below) emulates the ranks on one GPU.
 *  - Errors: every call returns a status. EINVAL for bad arguments (nothing enqueued),
 *    including a "device" buffer the GPU cannot dereference (pageable host memory;
 *    device, managed and pinned host memory are accepted — cudaPointerGetAttributes);
 *    ENOMEM when a call cannot allocate its working memory (the z-slab forward-projection
 *    array, host-path staging buffers): the call has not changed f or the context's images
 *    and the context stays usable; ECUDA/ENCCL for runtime failures (message in
 *    lmosem_last_error), after which the context answers ESTATE to everything except
 *    lmosem_last_error and lmosem_destroy.
 *  - Threading: one host thread per context; one context per GPU (rank).
 */
#ifndef LMOSEM_H
#define LMOSEM_H
#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef struct lmosem_ctx lmosem_ctx;

/* One list-mode event: a line of response between two detection points (mm). */
typedef struct {
    float x1, y1, z1, x2, y2, z2;
} lmosem_event;

typedef enum {
    LMOSEM_OK = 0,
    LMOSEM_EINVAL = 1,
    LMOSEM_ENOMEM = 2,
    LMOSEM_ECUDA = 3,
    LMOSEM_ENCCL = 4,
    LMOSEM_ESTATE = 5,
    LMOSEM_EIO = 6
} lmosem_status;

#define LMOSEM_NCCL_ID_BYTES 128

/* Multi-GPU setup; pass NULL for a single GPU without NCCL. nccl_unique_id points to
 * LMOSEM_NCCL_ID_BYTES bytes produced by lmosem_nccl_unique_id on one rank and broadcast
 * to all (the Python binding uses torch.distributed for the broadcast). A non-NULL dist
 * always creates the NCCL communicator and runs the combine (world == 1 included). */
typedef struct {
    int32_t rank, world;
    const void* nccl_unique_id;
} lmosem_dist;

/* Per-context counters. Phase times are summed CUDA-event durations (ms) on the
 * context's stream, recorded only while timing is enabled (lmosem_set_timing). */
typedef struct {
    int64_t launches;      /* kernels this context launched (all time) */
    int64_t subsets;       /* subset iterations completed (all time) */
    int64_t events;        /* events projected by this rank (all time) */
    int64_t timed_subsets; /* subsets covered by the phase times below */
    double convert_ms;     /* f -> internal brick layout (subset_step; first subset of reconstruct) */
    double project_ms;     /* step 1: fused traversal + forward + back-projection kernel */
    double combine_ms;     /* the combine (world > 1): ALLREDUCE the all-reduce of c; ISD the
                              reduce-scatter, the block update and the all-gather of f; FUSED
                              the fused kernel (which includes the block update) */
    double update_ms;      /* what follows the combine: ALLREDUCE (and one GPU) the step-2 update
                              kernel (also re-zeroes c); ISD / FUSED the brick -> caller-layout
                              copy of f (written on the last subset of a reconstruct) */
    double h2d_ms;         /* event uploads in lmosem_reconstruct_host (copy stream) */
    double tune_fused_ms;     /* world > 1: ms per combine of the fused kernel, of ISD and of */
    double tune_isd_ms;       /* ALLREDUCE, timed on this box at init (max over the ranks; */
    double tune_allreduce_ms; /* 0 = not timed), see lmosem_set_combine */
} lmosem_stats;

/* Library version as "lmosem <major>.<minor> sm_100a". */
const char* lmosem_version(void);

/* Block distribution: the event range [begin, end) of rank r of
 * world P for n events: begin = floor(r*n/P), end = floor((r+1)*n/P). Host only, no GPU
 * needed. EINVAL if n < 0, world < 1, rank outside [0, world) or a pointer is NULL. */
lmosem_status lmosem_block_range(int64_t n, int32_t rank, int32_t world, int64_t* begin, int64_t* end);

/* The ISD combine's brick blocks (the PSD -> ISD switch): the
 * internal image of n_bricks 8-float bricks is allocated as *alloc = n_bricks rounded up to a
 * multiple of world and split into world equal chunks; rank owns chunk `rank` (its part of
 * the reduce-scatter, the step-2 update and the all-gather), of which [*begin, *end) are real
 * bricks (*end <= n_bricks; a trailing chunk may be shorter or empty). Pure host function;
 * the blocks of ranks 0..world-1 partition [0, n_bricks). EINVAL on null pointers,
 * n_bricks < 0, world < 1 or rank outside [0, world). */
lmosem_status lmosem_isd_block(int64_t n_bricks, int32_t rank, int32_t world, int64_t* begin, int64_t* end,
                               int64_t* alloc);

/* Writes a fresh NCCL unique id (LMOSEM_NCCL_ID_BYTES bytes) to out. ENCCL on failure. */
lmosem_status lmosem_nccl_unique_id(void* out, size_t size);

/* Creates a context on the current CUDA device.
 *   dims[3]     = {nx, ny, nz} > 0, V < 2^31 (padded internal image < 2^31 floats), and
 *                 at most one extent > 1170: the per-warp path buffer (3 pieces per
 *                 dominant-axis slab) must fit in shared memory, so step 1 cuts a longer
 *                 axis into slabs of <= 1170 voxels (lmosem_set_slabs); EINVAL otherwise
 *   voxel_mm[3] = voxel size in mm, finite and > 0 (float64: the geometry is float64)
 *   norm        = V float32 sensitivity image s (device or host); copied, caller keeps it
 *   dist        = NULL for one GPU, else the rank/world/NCCL id (collective init;
 *                 EINVAL if world < 1, rank outside [0, world) or the id is NULL)
 * Returns EINVAL / ENOMEM / ECUDA / ENCCL; *out is NULL on failure. */
lmosem_status lmosem_init(lmosem_ctx** out, const int32_t dims[3], const double voxel_mm[3],
                          const float* norm, const lmosem_dist* dist);

/* Combine of the per-GPU error images (world > 1; needs a context created with a dist):
 *   LMOSEM_COMBINE_ALLREDUCE: ncclAllReduce(c), then every rank updates its full replica;
 *   LMOSEM_COMBINE_ISD: the paper's PSD -> ISD switch (Listing 3
 *     l.15-19): ncclReduceScatter(c) gives rank r the sum over its contiguous block of the
 *     internal image, rank r updates only that block (1/P of step 2), ncclAllGather
 *     rebuilds the full f on every rank. Same NVLink bytes, 1/P of the update work.
 * 0 (default) = for world > 1 over NCCL: the fused combine is set up and self-tested at
 * init, then it, ISD and ALLREDUCE are each timed on this box (lmosem_stats.tune_*_ms, max
 * over the ranks) and the fastest is the automatic combine (only ISD and ALLREDUCE are timed
 * when the fused one cannot be set up or fails its self-test); ISD with LMOSEM_AUTO_FUSED=0.
 * ALLREDUCE for world == 1. EINVAL for other values. */
#define LMOSEM_COMBINE_ALLREDUCE 1
#define LMOSEM_COMBINE_ISD 2
/* LMOSEM_COMBINE_FUSED (automatic for world > 1 when it passes its
 * self-test and times faster than ISD, see above): the ISD switch as ONE kernel over
 * NVLink peer memory (NCCL 2.28 symmetric windows + device communicator): rank r reads its
 * block of c summed over ranks (multimem.ld_reduce in the NVSwitch when available, else
 * peer loads), updates it and writes the new f block to every rank (multimem.st or peer
 * stores), between two LSA barriers. Setting it up runs a self-test of the kernel on a known
 * pattern on every rank (verdict agreed over the communicator; failure = ENCCL, the NCCL
 * collectives stay in use). Selecting it is COLLECTIVE (window registration); it
 * needs a context with a dist and all ranks in one NVLink domain, else ENCCL (not fatal,
 * the mode is unchanged, reason in lmosem_last_error). Its multi-rank logic is validated on
 * one GPU through the loopback transport below (the same kernel body); NCCL's LSA barriers,
 * windows and multimem run only on a multi-GPU NVLink node. */
#define LMOSEM_COMBINE_FUSED 3
lmosem_status lmosem_set_combine(lmosem_ctx* ctx, int32_t mode);

/* Emulated world (loopback transport, for tests on ONE GPU). A loopback group of `world`
 * ranks (1..16) stands in for an NCCL communicator: lmosem_init_loopback creates the
 * context of one rank on the current device (all ranks of a group on the same device, one
 * context per rank). The contexts then behave exactly like `world` NCCL ranks — collective
 * calls (subset_step, reconstruct*, sensitivity) must be made by every rank, each from its
 * own host thread — and run the same combine code: block split of
 * the events, the chosen combine (ALLREDUCE / ISD / FUSED; FUSED needs no set-up here), f
 * replicated. Each collective is NCCL-equivalent: sums over the ranks in rank order, made
 * by kernels that read the other ranks' buffers behind a host barrier plus stream events.
 * A rank that does not reach a collective within LMOSEM_TIMEOUT_S seconds (default 300)
 * fails it with ENCCL on every rank (the group is then broken). The group must outlive its
 * contexts: lmosem_loopback_destroy returns ESTATE while a context is still registered.
 * EINVAL: world outside 1..16, NULL pointers, rank outside [0, world), the rank already
 * taken, or a device other than the group's. */
typedef struct lmosem_loopback lmosem_loopback;
lmosem_status lmosem_loopback_create(int32_t world, lmosem_loopback** out);
lmosem_status lmosem_loopback_destroy(lmosem_loopback* group);
lmosem_status lmosem_init_loopback(lmosem_ctx** out, const int32_t dims[3], const double voxel_mm[3],
                                   const float* norm, lmosem_loopback* group, int32_t rank);

/* The combine mode in effect (-1 for a NULL context). */
int32_t lmosem_get_combine(const lmosem_ctx* ctx);

/* Out-of-L2 strategy: step 1 runs as z-slab passes when the
 * image is too large for L2 — pass A accumulates each event's forward projection over
 * slabs of the volume, pass B back-projects slab by slab with the complete fp — so each
 * launch touches one L2-sized image slab. n_slabs = 0 (default) picks the count from a
 * 72 MB-per-slab L2 budget (1 = single fused pass); n_slabs > 0 forces it (clamped to
 * nz/2). The slabs are cut along z, or along the axis longer than 1170 voxels, whose
 * slabs are then never longer than 1170 (at least that many slabs whatever is asked).
 * With 2-4 slabs and fewer than 2^31 events per call the passes are listed (the default,
 * LMOSEM_ZLIST=2): one classification kernel per subset sorts the events into per-launch
 * index lists. LORs inside one of the overlapping fine windows (about half a slab wide, fine
 * enough that the window's f and c fit L2 together) are projected by one fused pass over
 * their window; LORs inside one of the overlapping slab-wide windows by passes A and B over
 * that window; the others by passes A and B over only the slabs they cross. The lists take
 * 4 B x events x (slabs + windows) of device memory, allocated on first use and kept with
 * the context (C4, 10^7 events, 3 + 22 + 13 lists: 1.5 GB); if that allocation fails the
 * unlisted two-pass form runs instead (same result up to fp32 rounding).
 * The result is the same up to fp32 rounding. EINVAL if n_slabs < 0. */
lmosem_status lmosem_set_slabs(lmosem_ctx* ctx, int32_t n_slabs);

/* The z-slab count step 1 currently uses (-1 for a NULL context). */
int32_t lmosem_get_slabs(const lmosem_ctx* ctx);

/* Uses the given cudaStream_t (as void*) for all later device work; NULL means the CUDA
 * default stream (torch's default stream is NULL). Until this is called the context uses
 * its own non-blocking stream. The stream must belong to the context's device. */
lmosem_status lmosem_set_stream(lmosem_ctx* ctx, void* stream);

/* One subset iteration (step 1, combine, step 2) over n_events device events; f is the
 * V float32 device image, updated in place. Stream-ordered. n_events == 0 leaves f
 * unchanged (c stays 0). */
lmosem_status lmosem_subset_step(lmosem_ctx* ctx, const lmosem_event* events, int64_t n_events, float* f);

/* n_iterations passes over subsets l = 0..n_subsets-1 in order; subset l is
 * events[offsets[l], offsets[l+1]) (offsets: host, n_subsets+1 non-decreasing int64,
 * offsets[0] >= 0). events and f are device buffers. Stream-ordered. */
lmosem_status lmosem_reconstruct(lmosem_ctx* ctx, const lmosem_event* events, const int64_t* offsets,
                                 int32_t n_subsets, int32_t n_iterations, float* f);

/* As lmosem_reconstruct with HOST events and HOST f (in: f0, out: result). Uploads f,
 * streams each subset's events (this rank's block only) to the device on a copy stream,
 * double-buffered so the upload of subset l+1 overlaps the projection of subset l,
 * downloads f. Synchronous. */
lmosem_status lmosem_reconstruct_host(lmosem_ctx* ctx, const lmosem_event* events, const int64_t* offsets,
                                      int32_t n_subsets, int32_t n_iterations, float* f);

/* As lmosem_reconstruct with the events read from a list-mode file (Listing 2
 * lines 2-3, read_events per subset): `path` is a raw array of lmosem_event records
 * (24 B each, native-endian float32, no header); subset l is records
 * [offsets[l], offsets[l+1]). Each rank reads only its block of every subset with pread
 * into double-buffered pinned staging buffers (context-owned), so the file read and the
 * H2D copy of subset l+1 overlap the projection of subset l. f: V float32 DEVICE image
 * (in: f0, out: result). Synchronous. EIO if the file cannot be opened or read or is
 * shorter than offsets[n_subsets] records (the context stays usable after EIO). */
lmosem_status lmosem_reconstruct_file(lmosem_ctx* ctx, const char* path, const int64_t* offsets,
                                      int32_t n_subsets, int32_t n_iterations, float* f);

/* Step 1 only, for tests: c_out (V float32, device) <- error image of n_events device
 * events against device image f (c starts from 0; no combine, no update). */
lmosem_status lmosem_error_image(lmosem_ctx* ctx, const lmosem_event* events, int64_t n_events,
                                 const float* f, float* c_out);

/* Forward projection only, for tests: fp_out[i] = sum_j a_ij f_j (float32, device). */
lmosem_status lmosem_forward(lmosem_ctx* ctx, const lmosem_event* events, int64_t n_events,
                             const float* f, float* fp_out);

/* Sensitivity (norm) image over a set of LORs (the norm image of
 * BASELINE.json north_star): s_out_j = sum_i a_ij, the back-projection of ones with the
 * same exact traversal as step 1 (no forward projection). s_out: V float32 device,
 * x-fastest, overwritten. Collective with world > 1 (block split + all-reduce, every rank
 * gets the full image). Stream-ordered. */
lmosem_status lmosem_sensitivity(lmosem_ctx* ctx, const lmosem_event* events, int64_t n_events, float* s_out);

/* Replaces the context's norm image s (V float32, device or host; copied). Waits for the
 * copy, so the caller may release `norm` on return; later calls use the new s. EINVAL for
 * NULL. */
lmosem_status lmosem_set_norm(lmosem_ctx* ctx, const float* norm);

/* Step 2 only, for tests: f_j <- f_j*c_j/s_j where c_j > 0 and s_j > 0 (device f and c,
 * both V float32 x-fastest; the context's norm); c is re-zeroed. */
lmosem_status lmosem_update(lmosem_ctx* ctx, float* f, float* c);

/* Waits for all work enqueued by this context. Reports asynchronous kernel faults. With an
 * NCCL communicator it is a watchdog: ncclCommGetAsyncError is polled, and after
 * LMOSEM_TIMEOUT_S seconds (default 300) without completion — a peer rank that died or never
 * reached the collective — ENCCL is returned; the context then answers ESTATE and
 * lmosem_destroy aborts its communicator (ncclCommAbort) before releasing it. The
 * synchronous host/file reconstructions wait the same way. */
lmosem_status lmosem_synchronize(lmosem_ctx* ctx);

/* Enables (1) / disables (0) per-phase CUDA-event timing; enabling clears the times. */
lmosem_status lmosem_set_timing(lmosem_ctx* ctx, int32_t enable);

/* Resolves pending timing events (synchronizes) and copies the counters to *out. */
lmosem_status lmosem_get_stats(lmosem_ctx* ctx, lmosem_stats* out);

/* Releases everything the context owns (synchronizes first). NULL is a no-op. */
lmosem_status lmosem_destroy(lmosem_ctx* ctx);

/* Last error message of ctx ("" if none). With ctx == NULL: the message of the last
 * failed lmosem_init on the calling thread. */
const char* lmosem_last_error(const lmosem_ctx* ctx);

#ifdef __cplusplus
}
#endif
#endif
