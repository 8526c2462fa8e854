// lmosem_kernels.cuh — sm_100a kernels of the LM-OSEM subset iteration.
//
// Step 1 (Listing 2 lines 5-13) is ONE fused kernel per subset, k_project: a
// warp owns one line of response (LOR) at a time:
//   - work: warps claim batches of <= 32 events from a global counter; one lane per event
//     does the float64 setup — clip to the volume, dominant axis a (largest |du_a| in
//     voxel units), minor-axis positions at the first slab plane and slopes du_b/du_a,
//     du_c/du_a (|slope| <= 1) in Q24.40 fixed point — broadcast to the warp by shuffles;
//   - pass 1 (geometry): lane k takes slabs k, k+32, ... of the dominant axis, stepping
//     its minor positions by exactly 32 slopes (integer adds). Each minor axis crosses at
//     most one plane inside a slab, so a slab holds <= 3 pieces; up-moving axes are kept
//     mirrored so the distance to the next plane is the 40-bit fraction, converted to
//     float exactly (crossings in [0,1] carry ~1e-7 voxel absolute error wherever the slab
//     lies). The pieces (j, len) are compacted into the warp's shared-memory path buffer
//     in path order, and f is gathered for them in the same loop;
//   - forward projection (lines 9-10): a warp reduction of the gathered f*len gives fp;
//   - pass 2 (back-projection, lines 12-13): lane m reads piece m and issues
//     red.global.add.f32 of len/fp into c; lanes hold consecutive pieces of one path, so
//     they share 32-byte sectors of the brick layout below. c stays resident in L2.
// Internal image layout ("bricks"): the volume is padded by a halo (2 voxels low, >= 2
// high, even extents) and stored as 2x2x2 bricks of 8 floats = one 32-byte L2 sector;
// index J = Jx(px) + Jy(py) + Jz(pz) with J_axis(p) = M_axis*(p>>1) + m_axis*(p&1),
// (M, m) = (8, 1), (8*BX, 2), (8*BX*BY, 4). Rounding slivers that step one voxel past
// the volume land in the halo (f = 0 there, c ignored), so the hot loop has no range
// checks. Step 2 (lines 16-17 + norm) is k_update over bricks; it also re-zeroes c and
// writes the caller's x-fastest f.
#pragma once
#include <cuda_runtime.h>
#include <math_constants.h>
#include <stdint.h>

#include <type_traits>

namespace lmk {

constexpr int HALO_LO = 2;  // padded coordinate p = i + HALO_LO

struct GridGeom {
    int n[3];         // nx, ny, nz (real volume)
    int P[3];         // padded extents (even, >= n + 4)
    int A[3], B[3];   // brick index of padded coordinate p on axis k: A[k]*p + B[k]*(p & 1)
    int clo[3], chi[3];  // clip box in voxels: [0, n) except z = [zlo, zhi) of a z-slab pass
    double lo[3];     // volume lower corner (mm): -n*v/2
    double v[3];      // voxel size (mm)
    double inv_v[3];  // 1 / voxel size (1/mm)
    unsigned long long tex_fb;  // 1-D texture object over the brick f (MODE 5), 0 = none
};

// J_axis(p) = M*(p>>1) + m*(p&1) = (M/2)*p + (m - M/2)*(p&1), (M, m) = (8,1), (8BX,2), (8BX*BY,4)
__device__ __forceinline__ int bidx(int A, int B, int p) { return A * p + B * (p & 1); }

// Minor-axis positions are fixed point Q24.40 (int64, 2^-40 voxel): exact integer
// stepping w(k) = w0 + k*s, floor = w >> 40, fraction = low 40 bits. The slope error
// (<= 2^-41 per slab) accumulates to < 1e-9 voxel over 600 slabs.
constexpr int FIX_BITS = 40;
#ifndef LMK_APPEND2
#define LMK_APPEND2 0  // 1: path-buffer prefix from two ballots on n = v0 + v1 + v2 (A/B)
#endif

// Per-LOR traversal state (broadcast lane -> warp by shuffles; 14 registers). The piece
// lengths of the first and last slab (where the clip meets the plane crossings) come from
// lor_setup in float64, through the warp's shared-memory clip area (k_project).
struct Lor {
    long long wb0, wc0;  // minor-axis positions at the plane u_a = i0 (Q24.40 voxels, stored frame)
    long long sb, sc;    // their change per slab (stored frame: <= 0)
    float ab, ac;     // crossing offset in a slab: d = g * a (g: distance to the plane, Q.40)
    float lunit;      // mm of chord per unit of u_a
    int i0, ns;       // first slab index along a, number of slabs
    int code;         // bits 0-1: dominant axis a; 2-3: step of b (1: +1, 3: -1, 0: none); 4-5: c
};

// Warp-uniform constants derived from Lor::code and the grid once per LOR.
struct Walk {
    int mb, mc;       // -1 for a mirrored (up-moving) axis, else 0: voxel index = floor(w) ^ m
    float bb, bc;     // 0, or +inf for an axis without a step (no crossing)
    int Aa, Ba, Ab, Bb, Ac, Bc;  // brick index coefficients of axes a, b, c
    int Db0, Db1, Dc0, Dc1;      // index change of a step for an even / odd padded coordinate
};

template <class T>
__device__ __forceinline__ T sel3(const T (&v)[3], int i) {
    return i == 0 ? v[0] : (i == 1 ? v[1] : v[2]);
}

// Sets up the traversal of the segment p1 -> p2. Returns false if it contributes
// nothing (non-finite, zero length, misses the half-open volume).
// clip[0..2] / clip[3..5]: the three piece lengths (slab units) of the first / last slab in
// float64. There the clip (volume entry and exit, segment ends, slab-pass boundaries) meets
// the plane crossings, and a piece between a clip and a crossing must not be the difference
// of two rounded floats (a 3.7e-4-slab piece carried 1.5e-4 relative error that way).
// clo/chi: the launch's clip box (g.clo/g.chi, or a fused window's box in a listed launch).
__device__ __forceinline__ bool lor_setup(const float* __restrict__ ev, const GridGeom& g, const int (&clo)[3],
                                          const int (&chi)[3], Lor& L, float clip[6]) {
    double p1[3], d[3], u1[3], D[3], rD[3];
    bool ok = true;
#pragma unroll
    for (int k = 0; k < 3; ++k) {
        p1[k] = (double)ev[k];
        double p2 = (double)ev[3 + k];
        ok = ok && isfinite(p1[k]) && isfinite(p2);
        d[k] = p2 - p1[k];
        // voxel coordinate: by division on a stationary axis, whose voxel row (a LOR lying
        // in or near a voxel face) is then decided exactly as the oracle decides it,
        // floor((p - lo) / v) in float64 (reading S6); a moving axis only needs
        // the coordinate to rounding (1 ulp moves a crossing by ~1e-16 voxel)
        u1[k] = (p1[k] - g.lo[k]) * g.inv_v[k];
        if (d[k] == 0.0) u1[k] = (p1[k] - g.lo[k]) / g.v[k];
        D[k] = d[k] * g.inv_v[k];
    }
    if (!ok) return false;
    const double Lmm = sqrt(d[0] * d[0] + d[1] * d[1] + d[2] * d[2]);
    if (!(Lmm > 0.0)) return false;
    double amin = 0.0, amax = 1.0;
#pragma unroll
    for (int k = 0; k < 3; ++k) {
        const double lo = (double)clo[k], hi = (double)chi[k];
        rD[k] = 0.0;
        if (D[k] != 0.0) {
            const double r = 1.0 / D[k];
            rD[k] = r;
            double t0 = (lo - u1[k]) * r, t1 = (hi - u1[k]) * r;
            amin = fmax(amin, fmin(t0, t1));
            amax = fmin(amax, fmax(t0, t1));
        } else if (u1[k] < lo || u1[k] >= hi || p1[k] < g.lo[k] || p1[k] >= g.lo[k] + (double)g.n[k] * g.v[k]) {
            return false;  // parallel to axis k and outside (the volume test in mm as the oracle's)
        }
    }
    if (!(amax > amin)) return false;
    const double ax = fabs(D[0]), ay = fabs(D[1]), az = fabs(D[2]);
    const int a = (ax >= ay && ax >= az) ? 0 : ((ay >= az) ? 1 : 2);
    const int b = (a == 0) ? 1 : 0;
    const int c = (a == 2) ? 1 : 2;
    const double Da = sel3(D, a), u1a = sel3(u1, a);
    const double Db = sel3(D, b), Dc = sel3(D, c), u1b = sel3(u1, b), u1c = sel3(u1, c);
    double ua_in = u1a + amin * Da, ua_out = u1a + amax * Da;
    if (Da < 0.0) { double t = ua_in; ua_in = ua_out; ua_out = t; }
    int i0 = max((int)floor(ua_in), sel3(clo, a));
    int il = min((int)ceil(ua_out) - 1, sel3(chi, a) - 1);
    if (il < i0) return false;
    const double rDa = sel3(rD, a);  // 1 / Da from the clip (Da != 0: the dominant axis)
    const double sb = Db * rDa, sc = Dc * rDa;
    const double fx = (double)(1LL << FIX_BITS);
    // Guard: by the clip, the minor positions over the slab range lie in [0, n] up to
    // rounding; coordinates so large that float64 cannot resolve the clip (|p| ~ 1e20 mm)
    // would push them outside the 2-voxel halo (and the Q24.40 range) -> drop such LORs.
    {
        const double wbf = u1b + ((double)i0 - u1a) * sb, wbl = wbf + (double)(il + 1 - i0) * sb;
        const double wcf = u1c + ((double)i0 - u1a) * sc, wcl = wcf + (double)(il + 1 - i0) * sc;
        const double nb = (double)sel3(g.n, b), nc = (double)sel3(g.n, c);
        if (!(fmin(wbf, wbl) > -1.0 && fmax(wbf, wbl) < nb + 1.0 && fmin(wcf, wcl) > -1.0 &&
              fmax(wcf, wcl) < nc + 1.0))
            return false;
    }
    // stored frame: an axis moving up is mirrored, w' = -w - 2^-40, so every moving axis
    // moves down and its distance to the next plane is its fraction (the 2^-40 offset keeps
    // an exactly integral position inside its half-open voxel: distance = one voxel)
    {
        // floor decided in float64, fraction rounded to Q.40 below 1: a stationary axis
        // (s = 0: w = u1 exactly) keeps the oracle's voxel row
        auto fix = [fx](double u) {
            const double fl = floor(u);
            const long long q = min(__double2ll_rn((u - fl) * fx), (1LL << FIX_BITS) - 1);
            return (long long)fl * (1LL << FIX_BITS) + q;
        };
        const long long wb = fix(u1b + ((double)i0 - u1a) * sb);
        const long long wc = fix(u1c + ((double)i0 - u1a) * sc);
        const long long qb = __double2ll_rn(sb * fx), qc = __double2ll_rn(sc * fx);
        L.wb0 = sb > 0.0 ? -wb - 1 : wb;
        L.sb = sb > 0.0 ? -qb : qb;
        L.wc0 = sc > 0.0 ? -wc - 1 : wc;
        L.sc = sc > 0.0 ? -qc : qc;
    }
    // crossing inside a slab: distance g (Q.40 units) to the next plane in the direction
    // of travel, divided by |slope|: d = g * 2^-40 / |s| (no step: never, d = +inf)
    // 1/|s| = |Da / Db| from the clip's reciprocals (no further division)
    const double rb = fabs(Da * sel3(rD, b)), rc = fabs(Da * sel3(rD, c));
    L.ab = sb != 0.0 ? (float)(rb / fx) : 0.0f;
    L.ac = sc != 0.0 ? (float)(rc / fx) : 0.0f;
    L.lunit = (float)(Lmm * fabs(rDa));
    {
        // crossing offsets of the minor axes inside slab i from the exact plane positions, in
        // the conventions of the fixed-point walk (a position exactly on a plane belongs to
        // the voxel above it: an up-moving axis crosses one voxel later, a down-moving one at 0)
        const double fin = fmin(fmax(ua_in - (double)i0, 0.0), 1.0), fout = fmin(fmax(ua_out - (double)il, 0.0), 1.0);
        auto clip_pieces = [&](int i, double dlo, double dhi, float* out) {
            const double wb = u1b + ((double)i - u1a) * sb, wc = u1c + ((double)i - u1a) * sc;
            const double gb = wb - floor(wb), gc = wc - floor(wc);
            const double db = sb > 0.0 ? (1.0 - gb) * rb : (sb < 0.0 ? gb * rb : CUDART_INF);
            const double dc = sc > 0.0 ? (1.0 - gc) * rc : (sc < 0.0 ? gc * rc : CUDART_INF);
            const double q1 = fmin(fmax(fmin(db, dc), dlo), dhi), q2 = fmin(fmax(fmax(db, dc), dlo), dhi);
            out[0] = (float)(q1 - dlo);
            out[1] = (float)(q2 - q1);
            out[2] = (float)(dhi - q2);
        };
        const bool one = il == i0;
        clip_pieces(i0, fin, one ? fout : 1.0, clip);
        clip_pieces(il, one ? fin : 0.0, fout, clip + 3);
    }
    L.i0 = i0;
    L.ns = il - i0 + 1;
    L.code = a | (sb > 0.0 ? 4 : (sb < 0.0 ? 12 : 0)) | (sc > 0.0 ? 16 : (sc < 0.0 ? 48 : 0));
    return true;
}

__device__ __forceinline__ double shfl_d(double v, int src) {
    int lo = __double2loint(v), hi = __double2hiint(v);
    lo = __shfl_sync(0xffffffffu, lo, src);
    hi = __shfl_sync(0xffffffffu, hi, src);
    return __hiloint2double(hi, lo);
}

__device__ __forceinline__ long long shfl_ll(long long v, int src) {
    int lo = (int)(unsigned long long)v, hi = (int)((unsigned long long)v >> 32);
    lo = __shfl_sync(0xffffffffu, lo, src);
    hi = __shfl_sync(0xffffffffu, hi, src);
    return (long long)(((unsigned long long)(unsigned)hi << 32) | (unsigned)lo);
}

__device__ __forceinline__ Lor shfl_lor(const Lor& s, int src) {
    Lor L;
    L.wb0 = shfl_ll(s.wb0, src);
    L.wc0 = shfl_ll(s.wc0, src);
    L.sb = shfl_ll(s.sb, src);
    L.sc = shfl_ll(s.sc, src);
    L.ab = __shfl_sync(0xffffffffu, s.ab, src);
    L.ac = __shfl_sync(0xffffffffu, s.ac, src);
    L.lunit = __shfl_sync(0xffffffffu, s.lunit, src);
    L.i0 = __shfl_sync(0xffffffffu, s.i0, src);
    L.ns = __shfl_sync(0xffffffffu, s.ns, src);
    L.code = __shfl_sync(0xffffffffu, s.code, src);
    return L;
}

__device__ __forceinline__ Walk make_walk(const Lor& L, const GridGeom& g) {
    Walk W;
    const int a = L.code & 3, b = (a == 0) ? 1 : 0, c = (a == 2) ? 1 : 2;
    const int cb = (L.code >> 2) & 3, cc = (L.code >> 4) & 3;
    const int stb = (cb == 1) - (cb == 3), stc = (cc == 1) - (cc == 3);
    W.mb = -(stb > 0);
    W.mc = -(stc > 0);
    W.bb = cb ? 0.0f : CUDART_INF_F;
    W.bc = cc ? 0.0f : CUDART_INF_F;
    W.Aa = sel3(g.A, a); W.Ba = sel3(g.B, a);
    W.Ab = sel3(g.A, b); W.Bb = sel3(g.B, b);
    W.Ac = sel3(g.A, c); W.Bc = sel3(g.B, c);
    // J(p + st) - J(p) = st*A + B*((p + st)&1 - (p&1)) = st*A + B (p even), st*A - B (p odd)
    W.Db0 = stb ? stb * W.Ab + W.Bb : 0;
    W.Db1 = stb ? stb * W.Ab - W.Bb : 0;
    W.Dc0 = stc ? stc * W.Ac + W.Bc : 0;
    W.Dc1 = stc ? stc * W.Ac - W.Bc : 0;
    return W;
}

// The (up to) three pieces of slab k: j = brick index, l = chord length in units of the
// slab along the dominant axis (x lunit = mm; 0 for an empty piece).
struct Pieces {
    int j0, j1, j2;
    float l0, l1, l2;
};

// Slab k of the LOR; wb, wc = minor positions at its plane (Q24.40), Ja = brick index
// contribution of its dominant-axis coordinate (the caller steps all three exactly).
// floor (int) and fraction (float, exact conversion of the 40 fraction bits) of a
// stored-frame Q24.40 position; the fraction is the distance to the next plane crossed.
__device__ __forceinline__ float fix_split(long long w, int& fl) {
    const unsigned hi = (unsigned)((unsigned long long)w >> 32), lo = (unsigned)w;
    fl = (int)hi >> (FIX_BITS - 32);
    return __ull2float_rn(((unsigned long long)(hi & ((1u << (FIX_BITS - 32)) - 1u)) << 32) | lo);
}

// Brick index of padded coordinate p on one axis (A*p + B*(p&1)) and of p + step.
__device__ __forceinline__ void bidx2(int A, int B, int D0, int D1, int p, int& J0, int& J1) {
    const bool odd = p & 1;
    J0 = A * p + (odd ? B : 0);
    J1 = J0 + (odd ? D1 : D0);
}

// Slab k of the LOR; wb, wc = stored-frame minor positions at its plane, Ja = brick
// index contribution of its dominant-axis coordinate (the caller steps all three).
__device__ __forceinline__ Pieces slab_pieces(const Lor& L, const Walk& W, int k, long long wb, long long wc,
                                              int Ja) {
    int fb, fc;
    const float gb = fix_split(wb, fb), gc = fix_split(wc, fc);
    const int ib = fb ^ W.mb, ic = fc ^ W.mc;  // voxel indices (un-mirrored)
    const float db = fmaf(gb, L.ab, W.bb);  // crossing offsets along u_a in the slab
    const float dc = fmaf(gc, L.ac, W.bc);
    // no clip here: the first and last slab's lengths are replaced by their float64 values
    const float q1 = fminf(fminf(db, dc), 1.0f);  // db, dc >= 0
    const float q2 = fminf(fmaxf(db, dc), 1.0f);
    int Jb0, Jb1, Jc0, Jc1;
    bidx2(W.Ab, W.Bb, W.Db0, W.Db1, ib, Jb0, Jb1);  // halo offsets of b, c are in Ja
    bidx2(W.Ac, W.Bc, W.Dc0, W.Dc1, ic, Jc0, Jc1);
    // piece 0 before both crossings, piece 2 after both, piece 1 after the first one
    Pieces P;
    P.j0 = Ja + Jb0 + Jc0;
    P.j1 = Ja + ((db <= dc) ? (Jb1 + Jc0) : (Jb0 + Jc1));
    P.j2 = Ja + Jb1 + Jc1;
    // lengths in units of the slab (u_a); the LOR's mm per unit, lunit, is applied once per
    // LOR to fp and to the back-projected weight (three multiplies fewer per slab)
    P.l0 = q1;
    P.l1 = q2 - q1;
    P.l2 = 1.0f - q2;
    return P;
}

// Per-lane stepping state of a LOR's geometry loop: lane l visits slabs l, l+32, ...;
// positions advance by exactly 32 slopes (integer adds), so w(k) = w0 + k*s exactly.
struct Step {
    long long wb, wc, dwb, dwc;
    int Ja, dJa;
};

__device__ __forceinline__ Step make_step(const Lor& L, const Walk& W, int lane) {
    Step S;
    S.wb = L.wb0 + (long long)lane * L.sb;
    S.wc = L.wc0 + (long long)lane * L.sc;
    S.dwb = 32LL * L.sb;
    S.dwc = 32LL * L.sc;
    // 32 slabs later: same parity. HALO_LO is even, so J(i + HALO_LO) = J(i) + HALO_LO*A on
    // every axis: the minor axes' halo offsets are folded in here.
    S.Ja = bidx(W.Aa, W.Ba, L.i0 + lane + HALO_LO) + HALO_LO * (W.Ab + W.Ac);
    S.dJa = 32 * W.Aa;
    return S;
}

__device__ __forceinline__ void advance(Step& S) {
    S.wb += S.dwb;
    S.wc += S.dwc;
    S.Ja += S.dJa;
}

__device__ __forceinline__ float warp_sum(float v) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(0xffffffffu, v, o);
    return v;
}

// Loads event idx (6 floats) directly: three 8-byte streaming loads (fallback for event
// tiles that are not 16-byte aligned).
__device__ __forceinline__ void load_event(const float* __restrict__ events, int64_t idx, float ev[6]) {
    const float2* p = reinterpret_cast<const float2*>(events + 6 * idx);
    float2 a = __ldcs(p), b = __ldcs(p + 1), c = __ldcs(p + 2);
    ev[0] = a.x; ev[1] = a.y; ev[2] = b.x; ev[3] = b.y; ev[4] = c.x; ev[5] = c.y;
}

// Appends the valid pieces of every lane to the warp's path buffer in path order
// (lane-major = slab order, then piece order): the exclusive prefix of the per-lane
// counts n = v0 + v1 + v2 (0..3) comes from two ballots on its bits.
__device__ __forceinline__ void sts2(unsigned addr, int j, float l) {
    asm volatile("st.shared.v2.b32 [%0], {%1, %2};" ::"r"(addr), "r"(j), "r"(__float_as_int(l)) : "memory");
}

__device__ __forceinline__ int2 lds2(unsigned addr) {
    int2 v;
    asm volatile("ld.shared.v2.b32 {%0, %1}, [%2];" : "=r"(v.x), "=r"(v.y) : "r"(addr) : "memory");
    return v;
}

__device__ __forceinline__ float lds1(unsigned addr) {
    float v;
    asm volatile("ld.shared.f32 %0, [%1];" : "=f"(v) : "r"(addr) : "memory");
    return v;
}

// The record of a set-up LOR in the warp's LOR area in the z-slab passes: written by its
// setup lane, read by all 32 lanes with broadcast loads when the warp walks it (4 loads
// instead of the 16 shuffles of shfl_lor: C4 -1.3 %). wb0 wc0 | sb sc | ab ac lunit i0 |
// ns code clip0 clip1 | clip2..5. Not in the fused pass: its 4 CTAs per SM would need the
// 228 KB shared-memory carveout and leave the texture gathers 28 KB of L1 (C2 +17 %;
// DESIGN.md §7).
__device__ __forceinline__ void lor_store(unsigned a, const Lor& L, const float clip[6]) {
    asm volatile("st.shared.v2.b64 [%0], {%1, %2};" ::"r"(a), "l"(L.wb0), "l"(L.wc0) : "memory");
    asm volatile("st.shared.v2.b64 [%0], {%1, %2};" ::"r"(a + 16u), "l"(L.sb), "l"(L.sc) : "memory");
    asm volatile("st.shared.v4.b32 [%0], {%1, %2, %3, %4};" ::"r"(a + 32u), "f"(L.ab), "f"(L.ac), "f"(L.lunit),
                 "r"(L.i0)
                 : "memory");
    asm volatile("st.shared.v4.b32 [%0], {%1, %2, %3, %4};" ::"r"(a + 48u), "r"(L.ns), "r"(L.code), "f"(clip[0]),
                 "f"(clip[1])
                 : "memory");
    asm volatile("st.shared.v4.f32 [%0], {%1, %2, %3, %4};" ::"r"(a + 64u), "f"(clip[2]), "f"(clip[3]), "f"(clip[4]),
                 "f"(clip[5])
                 : "memory");
}

__device__ __forceinline__ Lor lor_load(unsigned a) {
    Lor L;
    asm volatile("ld.shared.v2.b64 {%0, %1}, [%2];" : "=l"(L.wb0), "=l"(L.wc0) : "r"(a) : "memory");
    asm volatile("ld.shared.v2.b64 {%0, %1}, [%2];" : "=l"(L.sb), "=l"(L.sc) : "r"(a + 16u) : "memory");
    asm volatile("ld.shared.v4.b32 {%0, %1, %2, %3}, [%4];"
                 : "=f"(L.ab), "=f"(L.ac), "=f"(L.lunit), "=r"(L.i0)
                 : "r"(a + 32u)
                 : "memory");
    asm volatile("ld.shared.v2.b32 {%0, %1}, [%2];" : "=r"(L.ns), "=r"(L.code) : "r"(a + 48u) : "memory");
    return L;
}

// path_s: 32-bit shared-window address of the warp's path buffer (8 B per piece).
__device__ __forceinline__ void append3(unsigned path_s, int& cnt, unsigned lt, const Pieces& P, bool v0, bool v1,
                                        bool v2) {
#if LMK_APPEND2
    // exclusive prefix over lanes of n = v0 + v1 + v2 (0..3) from two ballots on its bits
    const unsigned n = (unsigned)v0 + (unsigned)v1 + (unsigned)v2;
    const unsigned b0 = __ballot_sync(0xffffffffu, n & 1u), b1 = __ballot_sync(0xffffffffu, n & 2u);
    const unsigned a = path_s + 8u * (unsigned)(cnt + __popc(b0 & lt) + 2 * __popc(b1 & lt));
    cnt += __popc(b0) + 2 * __popc(b1);
#else
    // exclusive prefix over lanes of v0 + v1 + v2 from three predicate ballots
    const unsigned b0 = __ballot_sync(0xffffffffu, v0), b1 = __ballot_sync(0xffffffffu, v1),
                   b2 = __ballot_sync(0xffffffffu, v2);
    const unsigned a = path_s + 8u * (unsigned)(cnt + __popc(b0 & lt) + __popc(b1 & lt) + __popc(b2 & lt));
    cnt += __popc(b0) + __popc(b1) + __popc(b2);
#endif
    if (v0) sts2(a, P.j0, P.l0);
    if (v1) sts2(a + (v0 ? 8u : 0u), P.j1, P.l1);
    if (v2) sts2(a + (v0 ? 8u : 0u) + (v1 ? 8u : 0u), P.j2, P.l2);
}

#ifndef LMK_CTA_THREADS
#define LMK_CTA_THREADS 256  // 8 warps
#endif
#ifndef LMK_MIN_BLOCKS
#define LMK_MIN_BLOCKS 3     // CTAs per SM
#endif
#ifndef LMK_WIDE_CTA_THREADS
#define LMK_WIDE_CTA_THREADS 224  // CTA size of MODE 6 (the fused pass of large launches)
#endif
#ifndef LMK_WIDE_MIN_BLOCKS
#define LMK_WIDE_MIN_BLOCKS 4
#endif
#ifndef LMK_SLAB_CTA_THREADS
#define LMK_SLAB_CTA_THREADS 128  // CTA size of the z-slab passes (modes 2, 3)
#endif
#ifndef LMK_SLAB_MIN_BLOCKS
#define LMK_SLAB_MIN_BLOCKS 7  // CTAs per SM of the z-slab passes (modes 2, 3)
#endif
constexpr int PROJ_THREADS = LMK_CTA_THREADS;
// k_project's LOR area, per warp after all path buffers: per event of its claim, the 6
// float64-derived piece lengths of its first and last slab (24 B), and in the z-slab passes
// (modes 2, 3) also the 56 B of its Lor (lor_store: 80 B per event)
constexpr unsigned kLorRecBytes = 80;
__host__ __device__ constexpr bool lor_in_smem(int mode) { return mode == 2 || mode == 3; }
__host__ __device__ constexpr size_t lor_bytes_per_warp(int mode) { return 32u * (lor_in_smem(mode) ? kLorRecBytes : 24u); }
#ifndef LMK_PASSA_TEX
#define LMK_PASSA_TEX 0  // z-slab pass A gathers through the texture pipe (A/B; round 1: slower)
#endif
#ifndef LMK_LATE_WAIT
#define LMK_LATE_WAIT 1  // listed pass A / window launches wait for their predecessor at exit (A/B)
#endif
#ifndef LMK_GEOM_UNROLL
#define LMK_GEOM_UNROLL 0  // unroll of the geometry loop (0 = the compiler's choice, 2x)
#endif
constexpr int kGeomUnroll = LMK_GEOM_UNROLL > 0 ? LMK_GEOM_UNROLL : 1;
#ifndef LMK_SETUP_ONLY
#define LMK_SETUP_ONLY 0  // diagnostic builds only: skip the traversal (setup cost)
#endif
#ifndef LMK_TRACE
#define LMK_TRACE 0  // diagnostic builds only (tools/trace_tail.py): per-warp timeline
#endif
#if LMK_TRACE
constexpr int kTraceWarps = 16384;
// per warp: globaltimer at entry, at its first LOR, at exit; LORs processed; claims
__device__ unsigned long long g_trace[kTraceWarps * 5];
__device__ __forceinline__ unsigned long long gtimer() {
    unsigned long long t;
    asm volatile("mov.u64 %0, %globaltimer;" : "=l"(t));
    return t;
}
#endif
// Programmatic dependent launch (the host launches a kernel that directly follows another
// of the library's with programmaticStreamSerialization; without it both are no-ops):
// pdl_trigger lets the next kernel in the stream start launching its CTAs (they occupy
// an SM only as this kernel's CTAs leave it); pdl_wait blocks until every prerequisite
// grid has completed and its memory is visible. Each kernel waits before its first
// access to an image or per-event array that an earlier kernel writes or reads.
__device__ __forceinline__ void pdl_trigger() { asm volatile("griddepcontrol.launch_dependents;" ::: "memory"); }
__device__ __forceinline__ void pdl_wait() { asm volatile("griddepcontrol.wait;" ::: "memory"); }

template <int MODE>
constexpr int proj_min_blocks() {
    return (MODE == 2 || MODE == 3) ? LMK_SLAB_MIN_BLOCKS : (MODE == 6 ? LMK_WIDE_MIN_BLOCKS : LMK_MIN_BLOCKS);
}
template <int MODE>
constexpr int proj_threads() {
    return (MODE == 2 || MODE == 3) ? LMK_SLAB_CTA_THREADS : (MODE == 6 ? LMK_WIDE_CTA_THREADS : LMK_CTA_THREADS);
}
__host__ __device__ constexpr int proj_threads_of(int mode) {
    return (mode == 2 || mode == 3) ? LMK_SLAB_CTA_THREADS : (mode == 6 ? LMK_WIDE_CTA_THREADS : LMK_CTA_THREADS);
}

// Dynamic shared memory: per warp `cap` path pieces (int j, float len) packed as int2
// (<= 3 per dominant-axis slab of the launch's clip box; MODEs 1/2 keep no path: only the
// 32-event tile, 96 entries).
// MODE 0: fused forward + back-projection into cb (step 1, image resident in L2).
// MODE 1: forward projection only, fp[i] = fp (tests).
// MODE 2: z-slab pass A: fp[i] += forward projection of the part of LOR i in the slab.
// MODE 3: z-slab pass B: back-projection of the slab part of LOR i with the complete
//         fp[i] from pass A (events with fp <= 0 skipped).
// MODE 4: sensitivity image: back-projection of ones, cb_j += a_ij (no forward
//         projection).
// MODE 5: MODE 0 with the gathers of f through the texture pipe (tex1Dfetch on g.tex_fb),
//         the default for the fused pass when the brick f fits a 1-D linear texture.
// MODE 6: MODE 5 with 28 warps per SM (224 threads x 4 CTAs) instead of 24: large launches
//         (a whole C2 subset: -1.7 %); a rank's small share keeps MODE 5 (fewer, larger
//         claims per warp).
// MODEs 2/3 are the out-of-L2 strategy: each pass touches only one
// L2-sized slab of the image.
// A listed launch (the listed z-slab form) runs over the concatenation of the
// k_zclass lists list[0 .. nseg) (list l: lists + l * cap, length counts[l]; indices into
// `events` and `fp`), in order. box = 1: an event of segment s is clipped to [lo[s], hi[s])
// along `axis` instead of the launch's box (windows, or a coarse slab among windows).
constexpr int kMaxSeg = 16;
struct ListArg {
    const int* lists;
    const int* counts;
    long long cap;
    int nseg, axis, box;
    int entry_wait;  // pass B: wait for the predecessor at entry (the first pass B of a subset)
    int list[kMaxSeg], lo[kMaxSeg], hi[kMaxSeg];
};

// LIST (MODEs 2, 3, 5, 6): the launch runs over the listed events of `la` instead of [0, n).
template <int MODE, bool LIST = false>
__global__ void __launch_bounds__(proj_threads<MODE>(), proj_min_blocks<MODE>()) k_project(const float* __restrict__ events, int64_t n,
                                                             const float* __restrict__ fb, float* __restrict__ cb,
                                                             float* __restrict__ fp, GridGeom g, int cap,
                                                             unsigned long long* __restrict__ work, int batch,
                                                             int gdiv, ListArg la) {
    constexpr bool kGather = MODE <= 2 || MODE >= 5;  // forward projection in this launch
    constexpr bool kScatter = MODE == 0 || MODE >= 3;  // back-projection
    // gathers of f through the texture path (pass A too with LMK_PASSA_TEX, A/B builds only)
    constexpr bool kTex = MODE >= 5 || (MODE == 2 && LMK_PASSA_TEX);
    extern __shared__ __align__(16) int2 smem_path[];
    const int lane = threadIdx.x & 31;
    const int wib = threadIdx.x >> 5;
    const unsigned path_s = (unsigned)__cvta_generic_to_shared(smem_path + (size_t)wib * cap);
    constexpr bool kLorSmem = lor_in_smem(MODE);
    constexpr unsigned kRec = kLorSmem ? kLorRecBytes : 24u;  // bytes per event in the LOR area
    constexpr unsigned kClipOff = kLorSmem ? 56u : 0u;      // its clip lengths in the record
    // the warp's LOR area after all path buffers (lor_bytes_per_warp)
    const unsigned lor_w = (unsigned)__cvta_generic_to_shared(smem_path + (size_t)(blockDim.x >> 5) * cap) +
                           (unsigned)wib * (unsigned)lor_bytes_per_warp(MODE);
    const unsigned lt = (1u << lane) - 1u;
    // dynamic work distribution: each warp claims consecutive events from a global counter
    // (work[0]; zero at launch), so unequal LOR lengths and small per-rank subsets do not
    // leave idle warps. Guided claim sizes: `batch` (<= 32) while there is plenty of work,
    // then remaining / (gdiv * warps in the grid), even and >= 2 (claims stay
    // 16-byte aligned) — a 32-event claim takes a warp ~0.1 ms at C2, so fixed claims
    // left a tail of that length at the end of every launch
    const int64_t warps_in_grid = (int64_t)gridDim.x * (blockDim.x >> 5);
    int take = batch;
    // the list and its length were written before the previous launch started (k_zclass
    // precedes a plain launch), so they are read before griddepcontrol.wait. The host sized
    // the grid for all events; the claim sizes follow the list's length (lmosem.cu
    // launch_mode's rule with its defaults: first claims 32 halved while a warp would get
    // fewer than 4, >= 4; guided divisor 3 from 6 rounds of 32-event claims, else 2)
    // ends of the segments in the concatenation, and their clip planes (static indices here:
    // a dynamic index into the parameter array would copy it to the stack)
    __shared__ int s_segend[LIST ? kMaxSeg : 1], s_seglo[LIST ? kMaxSeg : 1], s_seghi[LIST ? kMaxSeg : 1],
        s_seglist[LIST ? kMaxSeg : 1];
    if (LIST) {
        int acc = 0;
#pragma unroll
        for (int q = 0; q < kMaxSeg; ++q) {
            if (q < la.nseg) acc += __ldg(la.counts + la.list[q]);
            if (threadIdx.x == 0) {
                s_segend[q] = acc;
                s_seglo[q] = la.lo[q];
                s_seghi[q] = la.hi[q];
                s_seglist[q] = la.list[q];
            }
        }
        __syncthreads();
        n = (int64_t)acc;
        take = 32;
        while (take > 4 && n < (int64_t)take * warps_in_grid * 4) take >>= 1;
        batch = take;
        gdiv = n >= 6 * 32 * warps_in_grid ? 3 : 2;
    }
    // claims, event tiles and the float64 setup of the first LORs overlap the previous
    // kernel's tail; pass B reads fp during setup, so it waits at once — the first listed
    // pass B of a subset before it lets its dependents launch, so that every later listed
    // launch starts after all of pass A has completed and may wait late (late_wait)
    // A listed pass A or window launch (late_wait) depends on no earlier listed launch of the
    // subset: it reads f (final before the plain launch that starts the sequence) and adds into
    // c and fp with atomics; a listed pass B after the first one starts only once every pass A
    // has completed (above). So they wait for their predecessor only before exiting, and
    // overlap its tail with real work. A launch's completion still implies its predecessor's,
    // so the first pass B and the kernel after the sequence see all of it complete.
    const bool late_wait = LIST && LMK_LATE_WAIT && !(MODE == 3 && la.entry_wait);
    bool dep_ready = MODE == 3 || late_wait;
    if (MODE == 3 && !late_wait) pdl_wait();
    pdl_trigger();
#if LMK_TRACE
    const int gw = blockIdx.x * (blockDim.x >> 5) + wib;
    unsigned long long tr_start = gtimer(), tr_first = 0, tr_lors = 0, tr_claims = 0;
#endif
    for (;;) {
        unsigned long long claim = 0;
        if (lane == 0) claim = atomicAdd(work, (unsigned long long)take);
        const int64_t base = (int64_t)__shfl_sync(0xffffffffu, claim, 0);
        if (base >= n) {
            // the last warp out re-zeroes the slot for the next launch (every other warp's
            // final claim returned before its exit count)
            if (lane == 0 && atomicAdd(work + 1, 1ull) == (unsigned long long)warps_in_grid - 1) {
                work[0] = 0;
                work[1] = 0;
            }
#if LMK_TRACE
            if (lane == 0 && gw < kTraceWarps) {
                unsigned long long* t = g_trace + 5 * gw;
                t[0] = tr_start; t[1] = tr_first; t[2] = gtimer(); t[3] = tr_lors; t[4] = tr_claims;
            }
#endif
            break;
        }
        const int64_t idx = base + lane;
        const bool mine_ev = lane < take && idx < n;
        // the event (and fp slot) of this lane: idx, or the idx-th listed event (segment sg)
        int64_t eidx = idx;
        int sg = 0;
        if (LIST) {
            eidx = 0;
            if (mine_ev) {
                int lo_i = 0;
                while (sg < la.nseg - 1 && idx >= s_segend[sg]) lo_i = s_segend[sg++];
                eidx = (int64_t)__ldg(la.lists + (int64_t)s_seglist[sg] * la.cap + (idx - lo_i));
            }
        }
        // event tile staging: the claimed events (24 B each, contiguous) are loaded with
        // coalesced 16-byte vector loads into the head of the warp's path buffer (idle at
        // this point), then each lane reads its record from shared memory
        const int m = (int)min((int64_t)take, n - base);
        if (gdiv > 0) {  // 0: fixed claims
            const int64_t rem = n - base - take;  // work left after this claim (estimate)
            const int64_t g = rem / (gdiv * warps_in_grid);
            take = batch <= 2 ? batch : (int)max((int64_t)2, min((int64_t)batch, g)) & ~1;
        }
        const float* tile_g = events + 6 * base;
        const bool vec = !LIST && ((((uintptr_t)tile_g) & 15) == 0) && ((m & 1) == 0);
        float4* tile_s = reinterpret_cast<float4*>(smem_path + (size_t)wib * cap);
        if (vec) {
            const float4* src = reinterpret_cast<const float4*>(tile_g);
            for (int q = lane; q < (3 * m) / 2; q += 32) tile_s[q] = __ldcs(src + q);
        }
        __syncwarp();
        Lor mine;
        bool ok = false;
        float fp_known = 1.0f;  // MODE 4 back-projects len * 1
        if (mine_ev) {
            float ev[6];
            if (vec) {
                const float2* r = reinterpret_cast<const float2*>(tile_s) + 3 * lane;
                const float2 a = r[0], b = r[1], c = r[2];
                ev[0] = a.x; ev[1] = a.y; ev[2] = b.x; ev[3] = b.y; ev[4] = c.x; ev[5] = c.y;
            } else {
                load_event(events, eidx, ev);
            }
            float clip[6];
            int clo[3], chi[3];
#pragma unroll
            for (int k = 0; k < 3; ++k) {
                const bool w = LIST && la.box && k == la.axis;
                clo[k] = w ? s_seglo[sg] : g.clo[k];
                chi[k] = w ? s_seghi[sg] : g.chi[k];
            }
            ok = lor_setup(ev, g, clo, chi, mine, clip);
            if (ok && kLorSmem) {
                lor_store(lor_w + kRec * (unsigned)lane, mine, clip);
            } else if (ok) {
                const unsigned a = lor_w + kRec * (unsigned)lane;
                asm volatile("st.shared.v2.f32 [%0], {%1, %2};" ::"r"(a), "f"(clip[0]), "f"(clip[1]) : "memory");
                asm volatile("st.shared.v2.f32 [%0], {%1, %2};" ::"r"(a + 8u), "f"(clip[2]), "f"(clip[3]) : "memory");
                asm volatile("st.shared.v2.f32 [%0], {%1, %2};" ::"r"(a + 16u), "f"(clip[4]), "f"(clip[5]) : "memory");
            }
            if (MODE == 3) {
                fp_known = fp[eidx];
                ok = ok && fp_known > 0.0f;  // reading S7
            }
        }
        if (!dep_ready) {  // warp-uniform
            pdl_wait();
            dep_ready = true;
        }
        if (MODE == 1 && mine_ev && !ok) fp[eidx] = 0.0f;
        __syncwarp();  // the tile is dead: the path buffer may be overwritten
        unsigned mask = __ballot_sync(0xffffffffu, ok);
#if LMK_SETUP_ONLY
        // diagnostic builds only (tools/ab_variants.py setup_only): claims, tiles and the
        // float64 setup without the traversal (the result is kept live, never stored)
        if (ok) {
            const unsigned h = (unsigned)mine.wb0 ^ (unsigned)mine.wc0 ^ (unsigned)mine.sb ^ (unsigned)mine.sc ^
                               __float_as_uint(mine.ab + mine.ac + mine.lunit) ^
                               (unsigned)(mine.i0 ^ mine.ns ^ mine.code);
            if (h == 0x9e3779b9u) cb[0] += 1.0f;
        }
        mask = 0;
#endif
#if LMK_TRACE
        tr_claims++;
        if (!tr_first && mask) tr_first = gtimer();
        tr_lors += __popc(mask);
#endif
        while (mask) {
            const int src = __ffs(mask) - 1;
            mask &= mask - 1;
            const unsigned rec = lor_w + kRec * (unsigned)src;
            const Lor L = kLorSmem ? lor_load(rec) : shfl_lor(mine, src);
            const Walk W = make_walk(L, g);
            // pass 1: geometry (uniform loop; lanes past the last slab drop their pieces)
            // -> path pieces in shared memory (when back-projecting) and f gathered in the
            // same loop (when forward-projecting)
            int cnt = 0;
            float acc = 0.0f;
            Step S = make_step(L, W, lane);
            // one 32-slab round: lane l takes slab k0 + l. The first round's lane 0 (slab 0)
            // and the last round's lane with slab ns - 1 take their float64 clip lengths; the
            // rounds are peeled so that the middle ones carry no clip test
            const unsigned clip_l = rec + kClipOff;
            auto round = [&](int k0, auto first, auto last) {
                const int k = k0 + lane;
                const bool in = k < L.ns;  // lanes past the last slab compute garbage, store nothing
                Pieces P = slab_pieces(L, W, k, S.wb, S.wc, S.Ja);
                if (decltype(first)::value && k == 0) {
                    P.l0 = lds1(clip_l);
                    P.l1 = lds1(clip_l + 4u);
                    P.l2 = lds1(clip_l + 8u);
                }
                if (decltype(last)::value && k == L.ns - 1) {
                    P.l0 = lds1(clip_l + 12u);
                    P.l1 = lds1(clip_l + 16u);
                    P.l2 = lds1(clip_l + 20u);
                }
                const bool v0 = in && P.l0 > 0.0f, v1 = in && P.l1 > 0.0f, v2 = in && P.l2 > 0.0f;
                if (kScatter) append3(path_s, cnt, lt, P, v0, v1, v2);
                if (kGather) {
                    if (kTex) {
                        // texel index through the texture pipe: the gathers leave the LSU data
                        // pipe to the REDs and the path buffer
                        acc = fmaf(v0 ? tex1Dfetch<float>(g.tex_fb, P.j0) : 0.f, P.l0, acc);
                        acc = fmaf(v1 ? tex1Dfetch<float>(g.tex_fb, P.j1) : 0.f, P.l1, acc);
                        acc = fmaf(v2 ? tex1Dfetch<float>(g.tex_fb, P.j2) : 0.f, P.l2, acc);
                    } else {
                        acc = fmaf(v0 ? __ldg(fb + P.j0) : 0.f, P.l0, acc);
                        acc = fmaf(v1 ? __ldg(fb + P.j1) : 0.f, P.l1, acc);
                        acc = fmaf(v2 ? __ldg(fb + P.j2) : 0.f, P.l2, acc);
                    }
                }
            };
            using T_ = std::true_type;
            using F_ = std::false_type;
            if (L.ns <= 32) {
                round(0, T_(), T_());
            } else {
                round(0, T_(), F_());
                advance(S);
                int k0 = 32;
#if LMK_GEOM_UNROLL > 0
#pragma unroll (kGeomUnroll)
#endif
                for (; k0 + 32 < L.ns; k0 += 32, advance(S)) round(k0, F_(), F_());
                round(k0, F_(), T_());
            }
            float fpv = fp_known;
            if (kGather) {
                fpv = warp_sum(acc) * L.lunit;
                const int64_t esrc = LIST ? (int64_t)__shfl_sync(0xffffffffu, (int)eidx, src) : base + src;
                if (MODE == 1 && lane == 0) fp[esrc] = fpv;
                if (MODE == 2 && lane == 0) {
                    if (late_wait)
                        atomicAdd(fp + esrc, fpv);  // pass A launches of a LOR's slabs may overlap
                    else
                        fp[esrc] += fpv;
                }
            } else {
                fpv = __shfl_sync(0xffffffffu, fp_known, src);
            }
            __syncwarp();
            if (kScatter && fpv > 0.0f) {  // reading S7: skip events with fp <= 0
                // pass 2: back-projection, lane m <- piece m (path order: consecutive
                // lanes share 32-byte brick sectors)
                const float inv = L.lunit / fpv;
#pragma unroll 8
                for (int m = lane; m < cnt; m += 32) {
                    const int2 q = lds2(path_s + 8u * (unsigned)m);
                    atomicAdd(cb + q.x, __int_as_float(q.y) * inv);
                }
            }
            __syncwarp();
        }
    }
    if (late_wait) pdl_wait();
}

// ------------------------------------------------------------ listed z-slab form (C4)
// When the image exceeds L2 the projection runs slab by slab (MODEs 2, 3). k_zclass sorts
// each event of the subset, once, into the launches that need it ("Listed
// z-slab form"). The slab-axis range [zl, zh] of its chord clipped to the volume (float32
// against a grown box, zclass_bits) decides:
//   - inside fine window j (the first one), kZMarginF voxels clear of its planes: fine list
//     F_j. Such a LOR's pieces are those of the whole-volume clip, so one fused launch
//     (MODE 5/6) over the window's box projects it completely; a window's f and c fit L2
//     together. Windows may overlap (stride < width: more LORs fit one);
//   - else: coarse list X_k of every coarse slab k that [zl - m, zh + m] meets (passes A
//     and B over slab k; a listed LOR that misses the slab is dropped by its clip).
// An event that cannot contribute (non-finite, zero length, missing the volume) is in no
// list. Lists: lists + l * cap, lengths counts[l]; l < K coarse, K <= l < K + Kf fine.
constexpr int kZMaxLists = 64;
struct ZClass {
    int K, Kf, Km, axis;
    int cb[kZMaxLists + 1];  // coarse slab planes (voxels along axis): cb[0] = 0 .. cb[K] = n
    int wlo[kZMaxLists], whi[kZMaxLists];  // fine windows [wlo, whi): wlo = j * ws (the last
    float ws, ww, wlast;                   // one: wlast), whi = wlo + ww
    float ms, mw, mlast;                   // medium windows (coarse-slab wide), the same way
};

// The window of a family (starts j * stride, the last one at `last`; width w; cnt windows)
// that holds [zl, zh] kZMarginF clear of its planes, or -1. The window starting last at or
// below zl - m is the only candidate (earlier ones end earlier), besides the clamped last one.
__device__ __forceinline__ int win_fit(float zl, float zh, float m, float stride, float w, float last, int cnt) {
    if (cnt <= 0) return -1;
    const int j = min((int)floorf(fmaxf(zl - m, 0.0f) / stride), cnt - 1);
    const float lo = j == cnt - 1 ? last : (float)j * stride;
    if (zl >= lo + m && zh <= lo + w - m) return j;
    if (j > 0 && j == cnt - 1) {  // the last window may start below the stride grid
        const float lo2 = (float)(j - 1) * stride;
        if (zl >= lo2 + m && zh <= lo2 + w - m) return j - 1;
    }
    return -1;
}

// The lists of one event, as a code (first list << 4) | count (0: none): one window list, or
// the contiguous run of coarse slabs its range meets. Decided in float32 against a
// box grown by kZMarginF voxels, so the clipped range contains the float64 one (lor_setup)
// up to float32 rounding (< 1e-2 voxel while both ends lie within 2 volume extents of the
// centre; farther or non-finite LORs go to every coarse list, where lor_setup decides):
//   - a LOR is fine-local only kZMarginF clear of its window's planes;
//   - a coarse list gets every LOR whose grown range meets the slab (a superset);
//   - no list: clearly zero length or missing the grown box.
constexpr float kZMarginF = 0.02f;
__device__ __forceinline__ unsigned zlist_code(int first, int count) { return ((unsigned)first << 4) | (unsigned)count; }
__device__ __forceinline__ unsigned zclass_bits(const float ev[6], const GridGeom& g, const ZClass& zc) {
    constexpr float m = kZMarginF;
    const unsigned all = zlist_code(0, zc.K);
    const float nmax = (float)max(g.n[0], max(g.n[1], g.n[2]));
    float u1[3], D[3];
    bool far = false, zero = true;
#pragma unroll
    for (int k = 0; k < 3; ++k) {
        const float lo = (float)g.lo[k], iv = (float)g.inv_v[k], c = 0.5f * (float)g.n[k];
        const float a = (ev[k] - lo) * iv, b = (ev[3 + k] - lo) * iv;
        far = far || !(fabsf(a - c) <= 2.0f * nmax && fabsf(b - c) <= 2.0f * nmax);  // also NaN / inf
        zero = zero && ev[k] == ev[3 + k];
        u1[k] = a;
        D[k] = b - a;
    }
    if (far) return all;
    if (zero) return 0u;  // p1 == p2: zero length (exactly as lor_setup decides)
    float amin = 0.0f, amax = 1.0f;
#pragma unroll
    for (int k = 0; k < 3; ++k) {
        const float hi = (float)g.n[k] + m;
        if (ev[k] != ev[3 + k]) {
            // approximate reciprocal: its error (~1 ulp; 1/0 = inf drops the axis' bound)
            // only lengthens or shortens the grown clip far inside the margin
            float r;
            asm("rcp.approx.ftz.f32 %0, %1;" : "=f"(r) : "f"(D[k]));
            const float t0 = (-m - u1[k]) * r, t1 = (hi - u1[k]) * r;
            amin = fmaxf(amin, fminf(t0, t1));
            amax = fminf(amax, fmaxf(t0, t1));
        } else if (u1[k] < -m || u1[k] > hi) {
            return 0u;  // parallel to axis k, clearly outside
        }
    }
    if (!(amax >= amin)) return 0u;
    const float us = sel3(u1, zc.axis), Ds = sel3(D, zc.axis);
    const float za = fmaf(amin, Ds, us), zb = fmaf(amax, Ds, us);
    const float zl = fminf(za, zb), zh = fmaxf(za, zb);
    if (!isfinite(zl) || !isfinite(zh)) return all;
    const int jf = win_fit(zl, zh, m, zc.ws, zc.ww, zc.wlast, zc.Kf);
    if (jf >= 0) return zlist_code(zc.K + jf, 1);
    const int jm = win_fit(zl, zh, m, zc.ms, zc.mw, zc.mlast, zc.Km);
    if (jm >= 0) return zlist_code(zc.K + zc.Kf + jm, 1);
    int k0 = zc.K, k1 = -1;  // the coarse slabs met form one run
    for (int k = 0; k < zc.K; ++k)
        if (zh + m > (float)zc.cb[k] && zl - m < (float)zc.cb[k + 1]) {
            k0 = min(k0, k);
            k1 = k;
        }
    return k1 >= k0 ? zlist_code(k0, k1 - k0 + 1) : 0u;
}

// One CTA per chunk of kZChunk consecutive events (grid-stride): each event takes its slot in
// each of its (<= kZMaxBits) lists with a shared-memory atomic, then one global atomic per
// list and chunk reserves the chunk's range. (A global atomic per warp and list serialised on
// the list counters: 0.6-1.5 ms per C4 subset; warp ballots per list: 0.44 ms.) Within a
// list, events keep chunk order.
#ifndef LMK_ZPER
#define LMK_ZPER 4  // events per thread and chunk in k_zclass (A/B: 1 / 2 / 4 / 8 / 16: 161 / 137 / 138 / 194 / 358 us at C4)
#endif
constexpr int kZThreads = 256, kZPer = LMK_ZPER, kZChunk = kZThreads * kZPer;
constexpr int kZMaxBits = 4;  // lists per event: one window, or <= 4 coarse slabs (host: K <= 4)
__global__ void __launch_bounds__(kZThreads) k_zclass(const float* __restrict__ events, int64_t n, GridGeom g,
                                                      ZClass zc, int* __restrict__ lists, int64_t cap,
                                                      int* __restrict__ counts) {
    pdl_wait();
    pdl_trigger();
    __shared__ int s_cnt[kZMaxLists], s_base[kZMaxLists];
    const int nl = zc.K + zc.Kf + zc.Km;
    for (int64_t c0 = (int64_t)blockIdx.x * kZChunk; c0 < n; c0 += (int64_t)gridDim.x * kZChunk) {
        if ((int)threadIdx.x < nl) s_cnt[threadIdx.x] = 0;
        __syncthreads();
        unsigned bits[kZPer];
        // all kZPer events' loads in flight before the clips
        float ev[kZPer][6];
#pragma unroll
        for (int p = 0; p < kZPer; ++p) {
            const int64_t i = c0 + p * kZThreads + threadIdx.x;
            load_event(events, i < n ? i : n - 1, ev[p]);
        }
#pragma unroll
        for (int p = 0; p < kZPer; ++p)
            bits[p] = c0 + p * kZThreads + threadIdx.x < n ? zclass_bits(ev[p], g, zc) : 0u;
        int off[kZPer][kZMaxBits];
#pragma unroll
        for (int p = 0; p < kZPer; ++p) {
            const int l0 = (int)(bits[p] >> 4), cnt = (int)(bits[p] & 15u);
#pragma unroll
            for (int q = 0; q < kZMaxBits; ++q)
                if (q < cnt) off[p][q] = atomicAdd(&s_cnt[l0 + q], 1);
        }
        __syncthreads();
        if ((int)threadIdx.x < nl) s_base[threadIdx.x] = s_cnt[threadIdx.x] ? atomicAdd(counts + threadIdx.x, s_cnt[threadIdx.x]) : 0;
        __syncthreads();
#pragma unroll
        for (int p = 0; p < kZPer; ++p) {
            const int l0 = (int)(bits[p] >> 4), cnt = (int)(bits[p] & 15u);
            const int e = (int)(c0 + p * kZThreads + threadIdx.x);
#pragma unroll
            for (int q = 0; q < kZMaxBits; ++q)
                if (q < cnt) lists[(int64_t)(l0 + q) * cap + s_base[l0 + q] + off[p][q]] = e;
        }
        __syncthreads();  // s_cnt / s_base are rewritten by the next chunk
    }
}

// ---------------------------------------------------------------- brick <-> row layouts
// One thread per brick (8 voxels). Brick b = bx + BX*(by + BY*bz) holds padded voxels
// (2bx+dx, 2by+dy, 2bz+dz) at 8b + dx + 2dy + 4dz; real voxel i = p - HALO_LO.
struct BrickIt {
    int BX, BY, BZ;
    int64_t nb;
    int rhi[3];  // bricks [HALO_LO/2, rhi[k]) of axis k hold real voxels (0: no halo skipping)
};

// A brick with at least one real voxel (the fused combine skips halo-only bricks: their f
// stays 0 and nothing reads their c).
__device__ __forceinline__ bool real_brick(const BrickIt& it, int64_t b) {
    if (it.rhi[0] == 0) return true;
    const unsigned u = (unsigned)b, bx = u % (unsigned)it.BX, t = u / (unsigned)it.BX;
    const unsigned by = t % (unsigned)it.BY, bz = t / (unsigned)it.BY;
    constexpr unsigned lo = HALO_LO / 2;
    return bx >= lo && bx < (unsigned)it.rhi[0] && by >= lo && by < (unsigned)it.rhi[1] && bz >= lo &&
           bz < (unsigned)it.rhi[2];
}

__device__ __forceinline__ bool real_voxel(const GridGeom& g, int px, int py, int pz, int64_t& r) {
    const int ix = px - HALO_LO, iy = py - HALO_LO, iz = pz - HALO_LO;
    if ((unsigned)ix >= (unsigned)g.n[0] || (unsigned)iy >= (unsigned)g.n[1] || (unsigned)iz >= (unsigned)g.n[2])
        return false;
    r = (int64_t)ix + (int64_t)g.n[0] * ((int64_t)iy + (int64_t)g.n[1] * iz);
    return true;
}

// row (x-fastest, caller) -> bricks (halo = 0)
__global__ void __launch_bounds__(256) k_row_to_brick(const float* __restrict__ row, float* __restrict__ br,
                                                      GridGeom g, BrickIt it) {
    pdl_wait();
    pdl_trigger();
    for (int64_t b = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; b < it.nb; b += (int64_t)gridDim.x * blockDim.x) {
        const int bx = (int)(b % it.BX);
        const int64_t t = b / it.BX;
        const int by = (int)(t % it.BY), bz = (int)(t / it.BY);
        float v[8];
#pragma unroll
        for (int q = 0; q < 8; ++q) {
            int64_t r;
            v[q] = real_voxel(g, 2 * bx + (q & 1), 2 * by + ((q >> 1) & 1), 2 * bz + (q >> 2), r) ? __ldg(row + r) : 0.0f;
        }
        float4* o = reinterpret_cast<float4*>(br + 8 * b);
        o[0] = make_float4(v[0], v[1], v[2], v[3]);
        o[1] = make_float4(v[4], v[5], v[6], v[7]);
    }
}

// bricks -> row (real voxels only); optionally zeroes the bricks afterwards
__global__ void __launch_bounds__(256) k_brick_to_row(float* __restrict__ br, float* __restrict__ row, GridGeom g,
                                                      BrickIt it, int zero) {
    pdl_wait();
    pdl_trigger();
    for (int64_t b = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; b < it.nb; b += (int64_t)gridDim.x * blockDim.x) {
        const int bx = (int)(b % it.BX);
        const int64_t t = b / it.BX;
        const int by = (int)(t % it.BY), bz = (int)(t / it.BY);
        float4* p = reinterpret_cast<float4*>(br + 8 * b);
        const float4 a = p[0], c = p[1];
        const float v[8] = {a.x, a.y, a.z, a.w, c.x, c.y, c.z, c.w};
#pragma unroll
        for (int q = 0; q < 8; ++q) {
            int64_t r;
            if (real_voxel(g, 2 * bx + (q & 1), 2 * by + ((q >> 1) & 1), 2 * bz + (q >> 2), r)) row[r] = v[q];
        }
        if (zero) {
            p[0] = make_float4(0.f, 0.f, 0.f, 0.f);
            p[1] = make_float4(0.f, 0.f, 0.f, 0.f);
        }
    }
}

// Step 2: f_j <- f_j * c_j / s_j where c_j > 0 and s_j > 0 (reading S9), c_j <- 0.
// Updates the brick copy fb and writes the caller's row-layout f. Halo voxels keep
// fb = 0 (sb = 0 there, so the guard leaves them unchanged).
__device__ __forceinline__ float upd1(float f, float c, float s) {
    return (c > 0.0f && s > 0.0f) ? f * __fdiv_rn(c, s) : f;
}

// Bricks [b_begin, b_end) (the whole image, or this rank's block in the ISD combine).
// zero_to > 0 (ISD): the bricks of [0, zero_to) outside the block only get c <- 0 (the
// reduce-scatter left this rank's partial sums there), in the same launch.
__global__ void __launch_bounds__(256) k_update(float* __restrict__ fb, float* __restrict__ cb,
                                                const float* __restrict__ sb, float* __restrict__ f_row, GridGeom g,
                                                BrickIt it, int64_t b_begin, int64_t b_end, int64_t zero_to) {
    pdl_wait();
    pdl_trigger();
    const bool zero_rest = zero_to > 0;
    const int64_t v0 = zero_rest ? 0 : b_begin, v1 = zero_rest ? zero_to : b_end;
    for (int64_t b = v0 + (int64_t)blockIdx.x * blockDim.x + threadIdx.x; b < v1;
         b += (int64_t)gridDim.x * blockDim.x) {
        float4* F = reinterpret_cast<float4*>(fb + 8 * b);
        float4* C = reinterpret_cast<float4*>(cb + 8 * b);
        if (zero_rest && (b < b_begin || b >= b_end)) {
            C[0] = make_float4(0.f, 0.f, 0.f, 0.f);
            C[1] = make_float4(0.f, 0.f, 0.f, 0.f);
            continue;
        }
        const float4* S = reinterpret_cast<const float4*>(sb + 8 * b);
        float4 f0 = F[0], f1 = F[1];
        const float4 c0 = __ldcs(C), c1 = __ldcs(C + 1), s0 = __ldg(S), s1 = __ldg(S + 1);
        f0.x = upd1(f0.x, c0.x, s0.x); f0.y = upd1(f0.y, c0.y, s0.y);
        f0.z = upd1(f0.z, c0.z, s0.z); f0.w = upd1(f0.w, c0.w, s0.w);
        f1.x = upd1(f1.x, c1.x, s1.x); f1.y = upd1(f1.y, c1.y, s1.y);
        f1.z = upd1(f1.z, c1.z, s1.z); f1.w = upd1(f1.w, c1.w, s1.w);
        F[0] = f0;
        F[1] = f1;
        C[0] = make_float4(0.f, 0.f, 0.f, 0.f);
        C[1] = make_float4(0.f, 0.f, 0.f, 0.f);
        if (f_row) {
            const int bx = (int)(b % it.BX);
            const int64_t t = b / it.BX;
            const int by = (int)(t % it.BY), bz = (int)(t / it.BY);
            const float v[8] = {f0.x, f0.y, f0.z, f0.w, f1.x, f1.y, f1.z, f1.w};
#pragma unroll
            for (int q = 0; q < 8; ++q) {
                int64_t r;
                if (real_voxel(g, 2 * bx + (q & 1), 2 * by + ((q >> 1) & 1), 2 * bz + (q >> 2), r)) f_row[r] = v[q];
            }
        }
    }
}

// ------------------------------------------------------- fused ISD combine (NEXT-1) body
// The paper's PSD -> ISD switch (Listing 3 l.15-19) as one pass over
// peer memory, generic over the rank team T (lmosem_fused.cuh: the NCCL LSA team over NVLink;
// tests/cuda/combine_emu.cu: P emulated ranks on one GPU):
//   T::sync(k)              barrier of CTA k across the ranks (acquire-release)
//   T::rank(), T::size()
//   T::sum_c(off, c0, c1)   the brick at byte offset off of c, summed over the ranks
//   T::sum_c2(oa, ob, ...)  two bricks at once (loads of both in flight)
//   T::store_f(off, n0, n1) the new brick of f, written to every rank
// Rank q owns bricks [q*chunk, min((q+1)*chunk, nb)); CTA k of ctas strides over them.
__device__ __forceinline__ float4 add4(float4 a, float4 b) { return make_float4(a.x + b.x, a.y + b.y, a.z + b.z, a.w + b.w); }

__device__ __forceinline__ float4 upd4(float4 f, float4 c, float4 s) {
    return make_float4(upd1(f.x, c.x, s.x), upd1(f.y, c.y, s.y), upd1(f.z, c.z, s.z), upd1(f.w, c.w, s.w));
}

template <class T>
__device__ __forceinline__ void combine_fused_body(T team, int cta, int ctas, const float* __restrict__ sb,
                                                   float* __restrict__ c_local, const float* __restrict__ fb_local,
                                                   int64_t chunk, int64_t nb, const BrickIt& it) {
    team.sync(cta);  // every rank's projection has finished writing its c
    const int nr = team.size();
    const int64_t b0 = chunk * team.rank(), b1 = b0 + chunk < nb ? b0 + chunk : nb;
    const int64_t t0 = (int64_t)cta * blockDim.x + threadIdx.x, stride = (int64_t)ctas * blockDim.x;
    // two bricks per thread per iteration: their c sums are in flight together; halo-only
    // bricks are skipped (no exchange)
    int64_t b = b0 + t0;
    for (; b + stride < b1; b += 2 * stride) {
        const bool ra = real_brick(it, b), rb = real_brick(it, b + stride);
        const size_t oa = (size_t)b * 32, ob = (size_t)(b + stride) * 32;
        const float4* Fa = reinterpret_cast<const float4*>(fb_local + 8 * b);
        const float4* Fb = reinterpret_cast<const float4*>(fb_local + 8 * (b + stride));
        const float4* Sa = reinterpret_cast<const float4*>(sb + 8 * b);
        const float4* Sb = reinterpret_cast<const float4*>(sb + 8 * (b + stride));
        if (ra && rb) {
            float4 ca0, ca1, cb0, cb1;
            team.sum_c2(oa, ob, ca0, ca1, cb0, cb1);
            const float4 na0 = upd4(Fa[0], ca0, __ldg(Sa)), na1 = upd4(Fa[1], ca1, __ldg(Sa + 1));
            const float4 nb0 = upd4(Fb[0], cb0, __ldg(Sb)), nb1 = upd4(Fb[1], cb1, __ldg(Sb + 1));
            team.store_f(oa, na0, na1);
            team.store_f(ob, nb0, nb1);
        } else if (ra || rb) {
            const size_t off = ra ? oa : ob;
            const float4* F = ra ? Fa : Fb;
            const float4* S = ra ? Sa : Sb;
            float4 c0, c1;
            team.sum_c(off, c0, c1);
            team.store_f(off, upd4(F[0], c0, __ldg(S)), upd4(F[1], c1, __ldg(S + 1)));
        }
    }
    if (b < b1 && real_brick(it, b)) {
        const size_t off = (size_t)b * 32;
        float4 c0, c1;
        team.sum_c(off, c0, c1);
        const float4* F = reinterpret_cast<const float4*>(fb_local + 8 * b);
        const float4* S = reinterpret_cast<const float4*>(sb + 8 * b);
        const float4 n0 = upd4(F[0], c0, __ldg(S)), n1 = upd4(F[1], c1, __ldg(S + 1));
        team.store_f(off, n0, n1);
    }
    team.sync(cta);  // CTA k of every rank has read its bricks of every c and written f
    // re-zero, in the local c, exactly the bricks CTA k read on every rank (the barrier
    // orders CTA k across ranks, not the CTAs of one rank); halo-only bricks too (rounding
    // slivers of step 1 may have added to them; nobody reads them)
    float4* C = reinterpret_cast<float4*>(c_local);
    const float4 z = make_float4(0.f, 0.f, 0.f, 0.f);
    for (int q = 0; q < nr; ++q) {
        const int64_t q0 = chunk * q, q1 = q0 + chunk < nb ? q0 + chunk : nb;
        for (int64_t b = q0 + t0; b < q1; b += stride) {
            C[2 * b] = z;
            C[2 * b + 1] = z;
        }
    }
}

}  // namespace lmk
