/* lmgen.c — seeded synthetic list-mode PET input generator (see lmgen.h).
 * Input bytes only; no LM-OSEM arithmetic lives here. */
#include "lmgen.h"
#include <math.h>
#include <stddef.h>

#define LMGEN_MAX_ATTEMPTS 100000

static inline uint64_t mix64(uint64_t z) {
    z += 0x9E3779B97F4A7C15ull;
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
    return z ^ (z >> 31);
}

/* uniform in [0,1) from the counter (seed, event, attempt, draw) */
static inline double urand(uint64_t seed, int64_t ev, int64_t attempt, int draw) {
    uint64_t k = mix64(mix64(seed) ^ (uint64_t)ev);
    k = mix64(k ^ ((uint64_t)attempt << 8) ^ (uint64_t)draw);
    return (double)(k >> 11) * (1.0 / 9007199254740992.0);
}

static double activity(const lmgen_config* c, double x, double y, double z) {
    for (int s = 0; s < c->n_spheres; ++s) {
        const double* sp = c->spheres[s];
        double dx = x - sp[0], dy = y - sp[1], dz = z - sp[2];
        if (dx * dx + dy * dy + dz * dz <= sp[3] * sp[3]) return sp[4];
    }
    if (c->bg_kind == 0) {
        if (x * x + y * y <= c->bg_r * c->bg_r && fabs(z) <= c->bg_half_len) return c->bg_act;
    } else {
        if (x * x + y * y + z * z <= c->bg_r * c->bg_r) return c->bg_act;
    }
    return 0.0;
}

static double max_activity(const lmgen_config* c) {
    double m = c->bg_act;
    for (int s = 0; s < c->n_spheres; ++s)
        if (c->spheres[s][4] > m) m = c->spheres[s][4];
    return m;
}

/* Line through p with direction d leaves the square tube |x|,|y| <= h at parameter t>0.
 * Returns +inf when d has no x/y component. */
static double exit_t(double h, const double p[3], const double d[3]) {
    double t = INFINITY;
    for (int a = 0; a < 2; ++a) {
        if (d[a] > 0) { double ta = (h - p[a]) / d[a]; if (ta < t) t = ta; }
        else if (d[a] < 0) { double ta = (-h - p[a]) / d[a]; if (ta < t) t = ta; }
    }
    return t;
}

/* One attempt: 0 = accepted (writes out[6]), 1 = rejected. */
static int attempt_event(const lmgen_config* c, double amax, int64_t ev, int64_t at, float* out) {
    double p[3];
    uint64_t sd = c->seed;
    if (c->hot_frac > 0 && urand(sd, ev, at, 0) < c->hot_frac) {
        double r = c->hot_r * cbrt(urand(sd, ev, at, 1));
        double ct = 2.0 * urand(sd, ev, at, 2) - 1.0, st = sqrt(fmax(0.0, 1.0 - ct * ct));
        double ph = 2.0 * M_PI * urand(sd, ev, at, 3);
        p[0] = r * st * cos(ph); p[1] = r * st * sin(ph); p[2] = r * ct;
    } else {
        double rx = c->bg_r, rz = (c->bg_kind == 0) ? c->bg_half_len : c->bg_r;
        for (int s = 0; s < c->n_spheres; ++s) { /* inserts may poke outside the background */
            const double* sp = c->spheres[s];
            double ex = fmax(fabs(sp[0]), fabs(sp[1])) + sp[3], ez = fabs(sp[2]) + sp[3];
            if (ex > rx) rx = ex;
            if (ez > rz) rz = ez;
        }
        p[0] = (2.0 * urand(sd, ev, at, 1) - 1.0) * rx;
        p[1] = (2.0 * urand(sd, ev, at, 2) - 1.0) * rx;
        p[2] = (2.0 * urand(sd, ev, at, 3) - 1.0) * rz;
        if (urand(sd, ev, at, 4) * amax >= activity(c, p[0], p[1], p[2])) return 1;
    }
    double d[3];
    if (c->dir_mode == 0) {
        double ct = 2.0 * urand(sd, ev, at, 5) - 1.0, st = sqrt(fmax(0.0, 1.0 - ct * ct));
        double ph = 2.0 * M_PI * urand(sd, ev, at, 6);
        d[0] = st * cos(ph); d[1] = st * sin(ph); d[2] = ct;
    } else {
        double ct = c->cos_lo + (c->cos_hi - c->cos_lo) * urand(sd, ev, at, 5);
        if (urand(sd, ev, at, 7) < 0.5) ct = -ct;
        double st = sqrt(fmax(0.0, 1.0 - ct * ct));
        double k = floor(4.0 * urand(sd, ev, at, 6));
        double ph = (45.0 + 90.0 * k + c->az_jitter_deg * (2.0 * urand(sd, ev, at, 8) - 1.0)) * (M_PI / 180.0);
        d[0] = st * cos(ph); d[1] = st * sin(ph); d[2] = ct;
    }
    double tp = exit_t(c->h, p, d);
    double dm[3] = {-d[0], -d[1], -d[2]};
    double tm = exit_t(c->h, p, dm);
    if (!isfinite(tp) || !isfinite(tm)) return 1;
    double z2 = p[2] + tp * d[2], z1 = p[2] - tm * d[2];
    if (fabs(z1) > c->hz || fabs(z2) > c->hz) return 1;
    out[0] = (float)(p[0] - tm * d[0]); out[1] = (float)(p[1] - tm * d[1]); out[2] = (float)z1;
    out[3] = (float)(p[0] + tp * d[0]); out[4] = (float)(p[1] + tp * d[1]); out[5] = (float)z2;
    return 0;
}

int lmgen_events(const lmgen_config* cfg, int64_t first, int64_t count, float* out) {
    if (!cfg || !out || first < 0 || count < 0) return -1;
    double amax = max_activity(cfg);
    if (!(amax > 0) && !(cfg->hot_frac > 0)) return -1;
    int fail = 0;
#pragma omp parallel for schedule(static) reduction(| : fail)
    for (int64_t i = 0; i < count; ++i) {
        int64_t ev = first + i, at = 0;
        while (at < LMGEN_MAX_ATTEMPTS && attempt_event(cfg, amax, ev, at, out + 6 * i)) ++at;
        if (at == LMGEN_MAX_ATTEMPTS) fail = 1;
    }
    return fail ? -2 : 0;
}

/* Geometric acceptance at point p over K Fibonacci-sphere directions,
 * z_k = 1 - 2k/(K-1): with K odd the set contains the equatorial direction z = 0, which
 * always reaches both heads from inside the volume, so s > 0 everywhere. */
static double acceptance(const lmgen_config* c, const double p[3], int K) {
    const double ga = M_PI * (3.0 - sqrt(5.0));
    int hit = 0;
    for (int k = 0; k < K; ++k) {
        double z = (K > 1) ? 1.0 - 2.0 * k / (K - 1.0) : 0.0, r = sqrt(fmax(0.0, 1.0 - z * z));
        double d[3] = {r * cos(ga * k), r * sin(ga * k), z};
        double dm[3] = {-d[0], -d[1], -d[2]};
        double tp = exit_t(c->h, p, d), tm = exit_t(c->h, p, dm);
        if (!isfinite(tp) || !isfinite(tm)) continue;
        if (fabs(p[2] + tp * d[2]) <= c->hz && fabs(p[2] - tm * d[2]) <= c->hz) ++hit;
    }
    return (double)hit / K;
}

int lmgen_norm(const lmgen_config* cfg, float* out) {
    if (!cfg || !out || cfg->nx <= 0 || cfg->ny <= 0 || cfg->nz <= 0 || cfg->norm_dirs <= 0) return -1;
    const int64_t nx = cfg->nx, ny = cfg->ny, nz = cfg->nz;
    /* s is defined on |x|,|y|,|z| of the voxel centre: evaluate one octant, mirror. */
    const int64_t hx = (nx + 1) / 2, hy = (ny + 1) / 2, hzn = (nz + 1) / 2;
#pragma omp parallel for collapse(2) schedule(dynamic, 1)
    for (int64_t iz = 0; iz < hzn; ++iz)
        for (int64_t iy = 0; iy < hy; ++iy)
            for (int64_t ix = 0; ix < hx; ++ix) {
                double p[3] = {fabs((ix + 0.5 - nx / 2.0) * cfg->vx), fabs((iy + 0.5 - ny / 2.0) * cfg->vy),
                               fabs((iz + 0.5 - nz / 2.0) * cfg->vz)};
                float s = (float)acceptance(cfg, p, cfg->norm_dirs);
                int64_t xs[2] = {ix, nx - 1 - ix}, ys[2] = {iy, ny - 1 - iy}, zs[2] = {iz, nz - 1 - iz};
                for (int a = 0; a < 2; ++a)
                    for (int b = 0; b < 2; ++b)
                        for (int e = 0; e < 2; ++e)
                            out[xs[a] + nx * (ys[b] + ny * zs[e])] = s;
            }
    return 0;
}
