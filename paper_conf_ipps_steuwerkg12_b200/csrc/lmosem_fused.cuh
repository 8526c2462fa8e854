// lmosem_fused.cuh — §8(f) NEXT-1: the paper's PSD -> ISD switch (PAPER.md lines 509-518,
// Listing 3 l.15-19) as ONE kernel over NVLink peer memory (NCCL 2.28 device API):
//   barrier (every rank's projection has finished writing its c)
//   -> rank r reads its brick block of c summed over all ranks (multimem.ld_reduce through
//      the NVSwitch when the LSA team has multimem, else loads from every peer's window)
//   -> step 2 on the block (f*c/s guarded)
//   -> the new f block is written to every rank's brick f (multimem.st, else peer stores)
//   -> barrier (CTA k of every rank done) -> each CTA re-zeroes, in its local c, exactly
//      the bricks CTA k read on every rank (the LSA barrier orders CTA k across ranks,
//      not the CTAs of one rank, so no CTA may touch bricks another CTA still reads).
// Replaces reduce-scatter + update + all-gather by one kernel. NVLink bytes per GPU: the
// NVSwitch still pulls every rank's partial c of the block, so each GPU's egress for the
// reduce is ~(P-1)/P*|c| (23.6 MB of the 27 MB brick c at P = 8, >= 31 us at the ~770 GB/s
// peer rate); what multimem saves is the all-gather egress (one multimem.st per brick
// instead of P-1 stores) and the overlap of egress with ingress in one pass. Halo-only
// bricks (6.5 % of the C2 image) are not exchanged. Launched as a programmatic dependent
// launch after the projection (pdl_wait before the first barrier) and triggering its own
// dependents at once, so the next subset's k_project can claim events and run its float64
// setup during the combine (every CTA of this kernel is resident before any dependent CTA).
// The multi-rank logic runs on one GPU through the loopback transport (lmosem_loop.cuh,
// the same body with P emulated ranks); NCCL's LSA barrier, windows and multimem only on
// a multi-GPU node.
#pragma once
#include <cuda/atomic>
#include <nccl.h>
#include <nccl_device.h>

#include "lmosem_kernels.cuh"

namespace lmk {

__device__ __forceinline__ float4 mm_ld_reduce4(const float* p) {
    float4 v;
    asm volatile("multimem.ld_reduce.relaxed.sys.global.add.v4.f32 {%0,%1,%2,%3}, [%4];"
                 : "=f"(v.x), "=f"(v.y), "=f"(v.z), "=f"(v.w)
                 : "l"(p)
                 : "memory");
    return v;
}

__device__ __forceinline__ void mm_st4(float* p, float4 v) {
    asm volatile("multimem.st.relaxed.sys.global.v4.f32 [%0], {%1,%2,%3,%4};" ::"l"(p), "f"(v.x), "f"(v.y), "f"(v.z),
                 "f"(v.w)
                 : "memory");
}

// The NCCL LSA team (one NVLink domain) for combine_fused_body: symmetric windows over c
// and the brick f; multimem (NVLS, in-switch reduction) when the team has it, else loads
// and stores to every peer's window.
template <bool MM>
struct NcclTeam {
    ncclDevComm dc;
    ncclWindow_t wc, wf;
    __device__ __forceinline__ void sync(int k) {
        ncclLsaBarrierSession<ncclCoopCta> bar(ncclCoopCta(), dc, ncclTeamTagLsa(), k, MM);
        bar.sync(ncclCoopCta(), cuda::memory_order_acq_rel);
    }
    __device__ __forceinline__ int rank() const { return dc.lsaRank; }
    __device__ __forceinline__ int size() const { return dc.lsaSize; }
    __device__ __forceinline__ void sum_c(size_t off, float4& c0, float4& c1) {
        if (MM) {
            const float* pc = (const float*)ncclGetLsaMultimemPointer(wc, off, dc);
            c0 = mm_ld_reduce4(pc);
            c1 = mm_ld_reduce4(pc + 4);
        } else {
            c0 = make_float4(0.f, 0.f, 0.f, 0.f);
            c1 = c0;
            for (int p = 0; p < dc.lsaSize; ++p) {
                const float4* pc = (const float4*)ncclGetLsaPointer(wc, off, p);
                c0 = add4(c0, pc[0]);
                c1 = add4(c1, pc[1]);
            }
        }
    }
    __device__ __forceinline__ void sum_c2(size_t oa, size_t ob, float4& a0, float4& a1, float4& b0, float4& b1) {
        if (MM) {
            const float* pa = (const float*)ncclGetLsaMultimemPointer(wc, oa, dc);
            const float* pb = (const float*)ncclGetLsaMultimemPointer(wc, ob, dc);
            a0 = mm_ld_reduce4(pa);
            a1 = mm_ld_reduce4(pa + 4);
            b0 = mm_ld_reduce4(pb);
            b1 = mm_ld_reduce4(pb + 4);
        } else {
            a0 = make_float4(0.f, 0.f, 0.f, 0.f);
            a1 = a0;
            b0 = a0;
            b1 = a0;
            for (int p = 0; p < dc.lsaSize; ++p) {
                const char* base = (const char*)ncclGetLsaPointer(wc, 0, p);
                const float4* pa = (const float4*)(base + oa);
                const float4* pb = (const float4*)(base + ob);
                const float4 x0 = pa[0], x1 = pa[1], y0 = pb[0], y1 = pb[1];
                a0 = add4(a0, x0);
                a1 = add4(a1, x1);
                b0 = add4(b0, y0);
                b1 = add4(b1, y1);
            }
        }
    }
    __device__ __forceinline__ void store_f(size_t off, float4 n0, float4 n1) {
        if (MM) {
            float* pf = (float*)ncclGetLsaMultimemPointer(wf, off, dc);
            mm_st4(pf, n0);
            mm_st4(pf + 4, n1);
        } else {
            for (int p = 0; p < dc.lsaSize; ++p) {
                float4* pf = (float4*)ncclGetLsaPointer(wf, off, p);
                pf[0] = n0;
                pf[1] = n1;
            }
        }
    }
};

// One CTA per LSA barrier index.
template <bool MM>
__global__ void __launch_bounds__(256) k_combine_fused(ncclDevComm dc, ncclWindow_t wc, ncclWindow_t wf,
                                                       const float* __restrict__ sb, float* __restrict__ c_local,
                                                       const float* __restrict__ fb_local, int64_t chunk, int64_t nb,
                                                       BrickIt it) {
    pdl_wait();     // the projection of every CTA of this rank is complete
    pdl_trigger();  // all CTAs of this kernel are resident: the next kernel may start its prologue
    NcclTeam<MM> team{dc, wc, wf};
    combine_fused_body(team, blockIdx.x, gridDim.x, sb, c_local, fb_local, chunk, nb, it);
}

// Self-test of the fused combine on a known pattern (run once when it is set up, on every
// rank, before it may become the default): c = rank + 1, brick f = 1, s = 1 on every brick;
// afterwards every real brick must hold f = sum_q (q + 1) = P(P+1)/2 (exact in float32),
// every halo-only brick f = 1, and c = 0 everywhere.
__global__ void __launch_bounds__(256) k_selftest_fill(float* __restrict__ c, float* __restrict__ fb,
                                                       float* __restrict__ s, int64_t nbf, float cval) {
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < nbf; i += (int64_t)gridDim.x * blockDim.x) {
        c[i] = cval;
        fb[i] = 1.0f;
        s[i] = 1.0f;
    }
}

__global__ void __launch_bounds__(256) k_selftest_check(const float* __restrict__ c, const float* __restrict__ fb,
                                                        BrickIt it, float expect, int* __restrict__ bad) {
    int nbad = 0;
    for (int64_t b = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; b < it.nb; b += (int64_t)gridDim.x * blockDim.x) {
        const float e = real_brick(it, b) ? expect : 1.0f;
        for (int q = 0; q < 8; ++q) nbad += (fb[8 * b + q] != e) + (c[8 * b + q] != 0.0f);
    }
    if (nbad) atomicAdd(bad, nbad);
}

}  // namespace lmk
