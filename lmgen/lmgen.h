/* lmgen.h — seeded synthetic list-mode PET input generator.
 *
 * This module produces INPUT BYTES only: list-mode events (lines of response, LORs)
 * and the sensitivity ("norm") image. It holds none of the LM-OSEM arithmetic
 * (no voxel traversal, no projection, no update); both the CPU oracle (oracle/) and
 * the CUDA path (paper_conf_ipps_steuwerkg12_b200/) consume what it writes.
 *
 * Workload shape follows the paper's application study (§IV.C, lines
 * 586-591: a 150x150x280 image, ~10^8 events in ~10^2 equal subsets, quadHIDAC PET
 * data). The quadHIDAC scanner is modelled as four planar detector heads at |x| = h
 * and |y| = h, |z| <= hz.
 *
 * Determinism: every random number is a counter-based hash of
 * (seed, event_id, attempt, draw), so event i is bit-identical for any thread count,
 * chunking or rank split.
 */
#ifndef LMGEN_H
#define LMGEN_H
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

#define LMGEN_MAX_SPHERES 8

typedef struct {
    /* image grid (used by the norm image only); volume centred on the origin, mm */
    int32_t nx, ny, nz;
    double vx, vy, vz;
    /* scanner: planar heads at |x| = h and |y| = h; detection only for |z| <= hz */
    double h, hz;
    /* background activity: kind 0 = cylinder (radius r, |z| <= half_len), 1 = sphere (r) */
    int32_t bg_kind;
    double bg_r, bg_half_len, bg_act;
    /* inserts: {cx, cy, cz, r, activity}; the first containing sphere sets the activity */
    int32_t n_spheres;
    double spheres[LMGEN_MAX_SPHERES][5];
    /* hot-spot mixture (skewed config): with probability hot_frac the emission point is
       uniform in a sphere of radius hot_r at the origin, otherwise drawn from the phantom */
    double hot_frac, hot_r;
    /* directions: mode 0 = isotropic; mode 1 = skewed: |cos(theta)| ~ U[cos_lo, cos_hi]
       (theta from the z axis), azimuth 45 deg + k*90 deg +- az_jitter_deg */
    int32_t dir_mode;
    double cos_lo, cos_hi, az_jitter_deg;
    uint64_t seed;
    /* number of Fibonacci-sphere directions for the norm image (odd: includes z = 0) */
    int32_t norm_dirs;
} lmgen_config;

/* Writes events [first, first+count) as 6 float32 each (x1,y1,z1,x2,y2,z2; mm) into out.
 * Returns 0 on success, -1 on bad arguments, -2 if an event exhausted its attempts. */
int lmgen_events(const lmgen_config* cfg, int64_t first, int64_t count, float* out);

/* Writes the norm (sensitivity) image, V = nx*ny*nz float32, x fastest. s_j is the
 * fraction of cfg->norm_dirs Fibonacci-sphere directions whose line through the centre
 * of voxel j reaches both heads within |z| <= hz (geometric acceptance). Returns 0/-1. */
int lmgen_norm(const lmgen_config* cfg, float* out);

#ifdef __cplusplus
}
#endif
#endif
