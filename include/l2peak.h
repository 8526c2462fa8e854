/* l2peak.h — builder-written microbenchmarks for the roofline denominators of the LM-OSEM projection
 * kernel: the rate of scattered 4-byte fp32 operations on an
 * image-sized buffer that sits in L2, the resource the back-projection
 * (red.global.add, Listing 2 lines 12-13) and the forward-projection gathers
 * (lines 9-10) are bound by. Not part of the LM-OSEM path.
 */
#ifndef L2PEAK_H
#define L2PEAK_H
#include <stdint.h>
#ifdef __cplusplus
extern "C" {
#endif

enum {
    L2PEAK_RED_RANDOM = 0,    /* fp32 red.global.add at uniformly random addresses */
    L2PEAK_LDG_RANDOM = 1,    /* fp32 gathers at uniformly random addresses */
    L2PEAK_PAIR_RANDOM = 2,   /* one gather + one red per op (the projection's mix) */
    L2PEAK_RED_RUN8 = 3,      /* red where each 8 lanes hit 8 consecutive floats */
    L2PEAK_PAIR_RUN8 = 4,     /* gather + red, 8-lane runs */
    L2PEAK_PAIR_WARP32 = 5,   /* gather + red, each warp on 32 consecutive floats (fully
                                 coalesced: the L2 peak for this op mix) */
    L2PEAK_STREAM5 = 6,       /* the update kernel's pattern streamed: read 3 arrays, write 2
                                 (float4, 20 B per element); ops = elements x passes */
    L2PEAK_LDG_WARP32 = 7,    /* gathers only, each warp on 32 consecutive floats (coalesced) */
    L2PEAK_RED_WARP32 = 8     /* reds only, each warp on 32 consecutive floats (coalesced) */
};

/* Runs `mode` on the current device over a buffer of n_floats floats (three for
 * STREAM5; device memory allocated and freed inside), ops_per_thread per thread on a full-occupancy grid, after
 * one warm-up launch. Writes the kernel time (ms, CUDA events) and the number of 4-byte
 * element operations (a pair counts as one op). Returns 0, or -1 on a CUDA error. */
int l2peak_run(int mode, int64_t n_floats, int32_t ops_per_thread, float* ms, double* ops);

#ifdef __cplusplus
}
#endif
#endif
