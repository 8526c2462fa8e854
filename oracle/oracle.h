/* oracle.h — plain float64 CPU LM-OSEM: the parity oracle.
 *
 * TEST INFRASTRUCTURE ONLY. Only tests/, __graft_entry__.smoke() and bench.py's
 * cpu_baseline / --impl reference legs may load or call this library. The product path
 * (paper_conf_ipps_steuwerkg12_b200/) never includes, links or imports anything here,
 * and this file shares no code, header, table or helper with it.
 *
 * What it computes (§IV, Listing 2; readings S1-S17 in DESIGN.md):
 *   for each subset l (fixed order):                        Listing 2 line 1
 *     c <- 0                                                reading S8
 *     for each event i:                                     line 5
 *       path = compute_path(event_i)                        line 7  (exact Siddon, S1)
 *       fp   = sum_m f[path[m].coord] * path[m].len         lines 9-10
 *       if fp > 0: c[path[m].coord] += path[m].len / fp     lines 12-13 (S7: skip fp <= 0)
 *     for each voxel j: if c_j > 0 and s_j > 0: f_j *= c_j / s_j     lines 16-17 + norm (S9)
 *
 * Geometry (readings S3-S6): the volume is nx*ny*nz voxels of vx*vy*vz mm, centred on the
 * origin; voxel (ix,iy,iz) is the half-open box [x0+ix*vx, x0+(ix+1)*vx) x ..., with
 * x0 = -nx*vx/2; linear index j = ix + nx*(iy + ny*iz). An event is 6 float32
 * (x1,y1,z1,x2,y2,z2) in mm: the segment p1 -> p2 (S2). All arithmetic is float64; the
 * fp32 input bytes are promoted exactly.
 */
#ifndef LMOSEM_ORACLE_H
#define LMOSEM_ORACLE_H
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef struct {
    int32_t nx, ny, nz;
    double vx, vy, vz;
} oracle_geom;

/* compute_path (Listing 2 line 7) by Siddon's method (merged plane-crossing parameters,
 * voxel of each interval from its midpoint, zero-length intervals dropped).
 * Writes up to cap (coord, len) pairs in traversal order p1 -> p2; returns the count,
 * or -1 if cap is too small. Returns 0 for a segment that misses the volume, has zero
 * length or non-finite coordinates. */
int64_t oracle_siddon_path(const oracle_geom* g, const double p1[3], const double p2[3],
                           int32_t* coord, double* len, int64_t cap);

/* Brute-force path for tiny volumes: for every voxel, the exact length of the segment
 * inside the closed voxel box (per-voxel slab clip, O(V)). Pairs in increasing coord.
 * Independent of oracle_siddon_path (pin P2). Returns count or -1 if cap too small. */
int64_t oracle_boxclip_path(const oracle_geom* g, const double p1[3], const double p2[3],
                            int32_t* coord, double* len, int64_t cap);

/* Forward projection fp_i = sum_j a_ij f_j for n events (Listing 2 lines 9-10). */
void oracle_forward(const oracle_geom* g, const float* events, int64_t n, const double* f, double* fp);

/* Error image (step 1, Listing 2 lines 5-13) for n events; c is zeroed first (S8). */
void oracle_error_image(const oracle_geom* g, const float* events, int64_t n, const double* f, double* c);

/* Sensitivity image s_j = sum_i a_ij over n LORs (the back-projection of ones; the norm
 * image of BASELINE.json north_star). s is zeroed first. */
void oracle_sensitivity(const oracle_geom* g, const float* events, int64_t n, double* s);

/* Image update (step 2, Listing 2 lines 16-17, with the norm of BASELINE.json north_star):
 * f_j <- f_j * c_j / s_j if c_j > 0 and s_j > 0, else unchanged (S9). */
void oracle_update(int64_t V, double* f, const double* c, const float* s);

/* One subset iteration: c <- 0, step 1, step 2. f is float64 in/out. Returns 0 or -1 (OOM). */
int oracle_subset_step(const oracle_geom* g, const float* events, int64_t n, const float* s, double* f);

/* Full reconstruction: n_iterations x (subsets l = 0..n_subsets-1 in order), subset l is
 * events[offsets[l], offsets[l+1]) (S12, S13). Returns 0 or -1. */
int oracle_reconstruct(const oracle_geom* g, const float* events, const int64_t* offsets,
                       int32_t n_subsets, int32_t n_iterations, const float* s, double* f);

/* OpenMP thread control (the oracle's loops over events run in parallel). */
void oracle_set_threads(int32_t n);
int32_t oracle_get_threads(void);

#ifdef __cplusplus
}
#endif
#endif
