// lmosem_kernels.cuh — sm_100a kernels of the LM-OSEM subset iteration.
//
// Step 1 (Listing 2 lines 5-13) is ONE fused kernel per subset: every warp
// owns one line of response (LOR) at a time and walks it as a set of independent slabs
// of its dominant axis:
//   - per LOR, in float64: clip to the volume, pick the dominant axis a (largest
//     |du_a| in voxel units), the minor-axis positions at the first slab plane and the
//     slopes du_b/du_a, du_c/du_a (|slope| <= 1);
//   - per slab i (lane k handles slabs k, k+32, ...): because |slope| <= 1 each minor
//     axis crosses at most one voxel plane inside the slab, so the slab holds at most
//     three path pieces; the minor position at the slab plane is one float64 FMA, and
//     the crossing points are computed in float32 relative to that plane (all values in
//     [0,1], so absolute error ~1e-7 voxel, independent of where the slab lies);
//   - pass 1 gathers f along the pieces (forward projection, Listing 2 lines 9-10),
//     a warp reduction gives fp; pass 2 recomputes the pieces and issues fp32
//     red.global.add of len/fp into c (back-projection, lines 12-13). c (25 MB at the
//     paper's 150x150x280) stays resident in the 126 MB L2.
// Step 2 (lines 16-17 + norm) is a vectorised streaming kernel that also re-zeroes c.
#pragma once
#include <cuda_runtime.h>
#include <math_constants.h>
#include <stdint.h>

namespace lmk {

struct GridGeom {
    int n[3];          // nx, ny, nz
    int stride[3];     // 1, nx, nx*ny
    double lo[3];      // volume lower corner (mm): -n*v/2
    double inv_v[3];   // 1 / voxel size (1/mm)
};

// Per-LOR traversal state, 21 x 32-bit words (broadcast lane -> warp by shuffles).
struct Lor {
    double wb0, wc0;   // minor-axis positions (voxel units) at the plane u_a = i0
    double sb, sc;     // du_b/du_a, du_c/du_a
    float isb, isc;    // 1/|sb|, 1/|sc| (+inf when the slope is 0)
    float lunit;       // mm of chord per unit of u_a
    float fin, fout;   // clip inside the first / last slab (local coordinate in [0,1])
    int i0, ns;        // first slab index along a, number of slabs
    int sa, sbs, scs;  // linear strides of axes a, b, c
    int nb, nc;        // extents of axes b, c
    int steps;         // bit0/1: sb >0/<0, bit2/3: sc >0/<0
};

// Register-resident pick of element i of a 3-array (avoids local-memory indexing).
template <class T>
__device__ __forceinline__ T sel3(const T (&v)[3], int i) {
    return i == 0 ? v[0] : (i == 1 ? v[1] : v[2]);
}

// Sets up the traversal of the segment p1 -> p2. Returns false if it contributes
// nothing (non-finite, zero length, misses the half-open volume).
__device__ __forceinline__ bool lor_setup(const float* __restrict__ ev, const GridGeom& g, Lor& L) {
    double p1[3], d[3], u1[3], D[3];
    bool ok = true;
#pragma unroll
    for (int k = 0; k < 3; ++k) {
        p1[k] = (double)ev[k];
        double p2 = (double)ev[3 + k];
        ok = ok && isfinite(p1[k]) && isfinite(p2);
        d[k] = p2 - p1[k];
        u1[k] = (p1[k] - g.lo[k]) * g.inv_v[k];
        D[k] = d[k] * g.inv_v[k];
    }
    if (!ok) return false;
    const double Lmm = sqrt(d[0] * d[0] + d[1] * d[1] + d[2] * d[2]);
    if (!(Lmm > 0.0)) return false;
    double amin = 0.0, amax = 1.0;
#pragma unroll
    for (int k = 0; k < 3; ++k) {
        if (D[k] != 0.0) {
            double r = 1.0 / D[k];
            double t0 = -u1[k] * r, t1 = ((double)g.n[k] - u1[k]) * r;
            amin = fmax(amin, fmin(t0, t1));
            amax = fmin(amax, fmax(t0, t1));
        } else if (u1[k] < 0.0 || u1[k] >= (double)g.n[k]) {
            return false;
        }
    }
    if (!(amax > amin)) return false;
    // dominant axis in voxel units
    const double ax = fabs(D[0]), ay = fabs(D[1]), az = fabs(D[2]);
    int a = (ax >= ay && ax >= az) ? 0 : ((ay >= az) ? 1 : 2);
    int b = (a == 0) ? 1 : 0;
    int c = (a == 2) ? 1 : 2;
    const double Da = sel3(D, a), u1a = sel3(u1, a);
    const double Db = sel3(D, b), Dc = sel3(D, c), u1b = sel3(u1, b), u1c = sel3(u1, c);
    double ua_in = u1a + amin * Da, ua_out = u1a + amax * Da;
    if (Da < 0.0) { double t = ua_in; ua_in = ua_out; ua_out = t; }
    const int na = sel3(g.n, a);
    int i0 = (int)floor(ua_in);
    int il = (int)ceil(ua_out) - 1;
    i0 = max(i0, 0);
    il = min(il, na - 1);
    if (il < i0) return false;
    const double rDa = 1.0 / Da;
    const double sb = Db * rDa, sc = Dc * rDa;
    L.sb = sb;
    L.sc = sc;
    L.wb0 = u1b + ((double)i0 - u1a) * sb;
    L.wc0 = u1c + ((double)i0 - u1a) * sc;
    L.isb = (sb != 0.0) ? (float)(1.0 / fabs(sb)) : CUDART_INF_F;
    L.isc = (sc != 0.0) ? (float)(1.0 / fabs(sc)) : CUDART_INF_F;
    L.lunit = (float)(Lmm * fabs(rDa));
    L.fin = fminf(fmaxf((float)(ua_in - (double)i0), 0.0f), 1.0f);
    L.fout = fminf(fmaxf((float)(ua_out - (double)il), 0.0f), 1.0f);
    L.i0 = i0;
    L.ns = il - i0 + 1;
    L.sa = sel3(g.stride, a);
    L.sbs = sel3(g.stride, b);
    L.scs = sel3(g.stride, c);
    L.nb = sel3(g.n, b);
    L.nc = sel3(g.n, c);
    L.steps = (sb > 0.0 ? 1 : 0) | (sb < 0.0 ? 2 : 0) | (sc > 0.0 ? 4 : 0) | (sc < 0.0 ? 8 : 0);
    return true;
}

__device__ __forceinline__ double shfl_d(double v, int src) {
    int lo = __double2loint(v), hi = __double2hiint(v);
    lo = __shfl_sync(0xffffffffu, lo, src);
    hi = __shfl_sync(0xffffffffu, hi, src);
    return __hiloint2double(hi, lo);
}

__device__ __forceinline__ Lor shfl_lor(const Lor& s, int src) {
    Lor L;
    L.wb0 = shfl_d(s.wb0, src);
    L.wc0 = shfl_d(s.wc0, src);
    L.sb = shfl_d(s.sb, src);
    L.sc = shfl_d(s.sc, src);
    L.isb = __shfl_sync(0xffffffffu, s.isb, src);
    L.isc = __shfl_sync(0xffffffffu, s.isc, src);
    L.lunit = __shfl_sync(0xffffffffu, s.lunit, src);
    L.fin = __shfl_sync(0xffffffffu, s.fin, src);
    L.fout = __shfl_sync(0xffffffffu, s.fout, src);
    L.i0 = __shfl_sync(0xffffffffu, s.i0, src);
    L.ns = __shfl_sync(0xffffffffu, s.ns, src);
    L.sa = __shfl_sync(0xffffffffu, s.sa, src);
    L.sbs = __shfl_sync(0xffffffffu, s.sbs, src);
    L.scs = __shfl_sync(0xffffffffu, s.scs, src);
    L.nb = __shfl_sync(0xffffffffu, s.nb, src);
    L.nc = __shfl_sync(0xffffffffu, s.nc, src);
    L.steps = __shfl_sync(0xffffffffu, s.steps, src);
    return L;
}

// The (up to) three pieces of slab k of a LOR: calls emit(j, len) for each piece of
// positive length whose voxel lies in the volume.
template <class Emit>
__device__ __forceinline__ void slab_pieces(const Lor& L, int k, Emit&& emit) {
    const double wb = fma((double)k, L.sb, L.wb0);
    const double wc = fma((double)k, L.sc, L.wc0);
    const double fbb = floor(wb), fcc = floor(wc);
    const int bb = (int)fbb, cc = (int)fcc;
    const float fb = (float)(wb - fbb), fc = (float)(wc - fcc);
    const int stb = (L.steps & 1) ? 1 : ((L.steps & 2) ? -1 : 0);
    const int stc = (L.steps & 4) ? 1 : ((L.steps & 8) ? -1 : 0);
    // local crossing positions in [0, inf) along u_a from the slab's lower plane
    const float db = (stb > 0) ? (1.0f - fb) * L.isb : ((stb < 0) ? fb * L.isb : CUDART_INF_F);
    const float dc = (stc > 0) ? (1.0f - fc) * L.isc : ((stc < 0) ? fc * L.isc : CUDART_INF_F);
    const float dlo = (k == 0) ? L.fin : 0.0f;
    const float dhi = (k == L.ns - 1) ? L.fout : 1.0f;
    const float x1 = fminf(db, dc), x2 = fmaxf(db, dc);
    const float q1 = fminf(fmaxf(x1, dlo), dhi);
    const float q2 = fminf(fmaxf(x2, dlo), dhi);
    const int ja = (L.i0 + k) * L.sa;
    const float s[3] = {dlo, q1, q2};
    const float e[3] = {q1, q2, dhi};
#pragma unroll
    for (int p = 0; p < 3; ++p) {
        const int ib = bb + ((s[p] >= db) ? stb : 0);
        const int ic = cc + ((s[p] >= dc) ? stc : 0);
        const float len = (e[p] - s[p]) * L.lunit;
        const bool ok = (e[p] > s[p]) && ((unsigned)ib < (unsigned)L.nb) && ((unsigned)ic < (unsigned)L.nc);
        emit(ok, ja + ib * L.sbs + ic * L.scs, len);
    }
}

__device__ __forceinline__ float warp_sum(float v) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(0xffffffffu, v, o);
    return v;
}

// Loads event idx (6 floats) of an AoS array: three 8-byte loads (24-byte records are
// 8-byte aligned); consecutive lanes read consecutive records (coalesced 768 B / warp).
__device__ __forceinline__ void load_event(const float* __restrict__ events, int64_t idx, float ev[6]) {
    const float2* p = reinterpret_cast<const float2*>(events + 6 * idx);
    float2 a = __ldcs(p), b = __ldcs(p + 1), c = __ldcs(p + 2);
    ev[0] = a.x; ev[1] = a.y; ev[2] = b.x; ev[3] = b.y; ev[4] = c.x; ev[5] = c.y;
}

// MODE 0: fused forward + back-projection into c (step 1).
// MODE 1: forward projection only, fp written to fp_out[i] (tests).
template <int MODE>
__global__ void __launch_bounds__(256) k_project(const float* __restrict__ events, int64_t n,
                                                 const float* __restrict__ f, float* __restrict__ c,
                                                 float* __restrict__ fp_out, GridGeom g) {
    const int lane = threadIdx.x & 31;
    const int64_t warp = (int64_t)blockIdx.x * (blockDim.x >> 5) + (threadIdx.x >> 5);
    const int64_t nwarps = (int64_t)gridDim.x * (blockDim.x >> 5);
    for (int64_t base = warp * 32; base < n; base += nwarps * 32) {
        const int64_t idx = base + lane;
        Lor mine;
        bool ok = false;
        if (idx < n) {
            float ev[6];
            load_event(events, idx, ev);
            ok = lor_setup(ev, g, mine);
        }
        if (MODE == 1 && idx < n && !ok) fp_out[idx] = 0.0f;
        unsigned mask = __ballot_sync(0xffffffffu, ok);
        while (mask) {
            const int src = __ffs(mask) - 1;
            mask &= mask - 1;
            const Lor L = shfl_lor(mine, src);
            float acc = 0.0f;
            for (int k = lane; k < L.ns; k += 32) {
                slab_pieces(L, k, [&](bool v, int j, float len) {
                    if (v) acc = fmaf(__ldg(f + j), len, acc);
                });
            }
            const float fp = warp_sum(acc);
            if (MODE == 1) {
                if (lane == 0) fp_out[base + src] = fp;
                continue;
            }
            if (!(fp > 0.0f)) continue;  // reading S7: skip events with fp <= 0
            const float inv = 1.0f / fp;
            for (int k = lane; k < L.ns; k += 32) {
                slab_pieces(L, k, [&](bool v, int j, float len) {
                    if (v) atomicAdd(c + j, len * inv);
                });
            }
        }
    }
}

// Step 2: f_j <- f_j * c_j / s_j where c_j > 0 and s_j > 0; c_j <- 0 (next subset).
__device__ __forceinline__ float upd1(float f, float c, float s) {
    return (c > 0.0f && s > 0.0f) ? f * __fdiv_rn(c, s) : f;
}

// vec = 1 when f, c and s are 16-byte aligned (float4 path), else scalar throughout.
__global__ void __launch_bounds__(256) k_update(float* __restrict__ f, float* __restrict__ c,
                                                const float* __restrict__ s, int64_t V, int vec) {
    const int64_t n4 = vec ? (V >> 2) : 0;
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    float4* f4 = reinterpret_cast<float4*>(f);
    float4* c4 = reinterpret_cast<float4*>(c);
    const float4* s4 = reinterpret_cast<const float4*>(s);
    const float4 z = make_float4(0.f, 0.f, 0.f, 0.f);
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n4; i += stride) {
        float4 fv = f4[i], cv = __ldcs(c4 + i), sv = __ldg(s4 + i);
        fv.x = upd1(fv.x, cv.x, sv.x);
        fv.y = upd1(fv.y, cv.y, sv.y);
        fv.z = upd1(fv.z, cv.z, sv.z);
        fv.w = upd1(fv.w, cv.w, sv.w);
        f4[i] = fv;
        c4[i] = z;
    }
    for (int64_t i = (n4 << 2) + (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < V; i += stride) {
        f[i] = upd1(f[i], c[i], s[i]);
        c[i] = 0.0f;
    }
}

}  // namespace lmk
