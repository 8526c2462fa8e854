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
// Replaces reduce-scatter + update + all-gather; NVLink bytes per GPU with multimem are
// ~2*|c|/P instead of ~2*(P-1)/P*|c|. Opt-in (LMOSEM_COMBINE_FUSED): with one GPU per test
// call only the 1-rank peer-pointer path can be exercised here.
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

__device__ __forceinline__ float4 add4(float4 a, float4 b) { return make_float4(a.x + b.x, a.y + b.y, a.z + b.z, a.w + b.w); }

__device__ __forceinline__ float4 upd4(float4 f, float4 c, float4 s) {
    return make_float4(upd1(f.x, c.x, s.x), upd1(f.y, c.y, s.y), upd1(f.z, c.z, s.z), upd1(f.w, c.w, s.w));
}

// One CTA per LSA barrier index. Rank q owns bricks [q*chunk, min((q+1)*chunk, nb)).
template <bool MM>
__global__ void __launch_bounds__(256) k_combine_fused(ncclDevComm dc, ncclWindow_t wc, ncclWindow_t wf,
                                                       const float* __restrict__ sb, float* __restrict__ c_local,
                                                       const float* __restrict__ fb_local, int64_t chunk, int64_t nb) {
    {
        ncclLsaBarrierSession<ncclCoopCta> bar(ncclCoopCta(), dc, ncclTeamTagLsa(), blockIdx.x, MM);
        bar.sync(ncclCoopCta(), cuda::memory_order_acq_rel);
    }
    const int nr = dc.lsaSize;
    const int64_t b0 = chunk * dc.lsaRank, b1 = b0 + chunk < nb ? b0 + chunk : nb;
    const int64_t t0 = (int64_t)blockIdx.x * blockDim.x + threadIdx.x, stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t b = b0 + t0; b < b1; b += stride) {
        const size_t off = (size_t)b * 32;
        float4 c0, c1;
        if (MM) {
            const float* pc = (const float*)ncclGetLsaMultimemPointer(wc, off, dc);
            c0 = mm_ld_reduce4(pc);
            c1 = mm_ld_reduce4(pc + 4);
        } else {
            c0 = make_float4(0.f, 0.f, 0.f, 0.f);
            c1 = c0;
            for (int p = 0; p < nr; ++p) {
                const float4* pc = (const float4*)ncclGetLsaPointer(wc, off, p);
                c0 = add4(c0, pc[0]);
                c1 = add4(c1, pc[1]);
            }
        }
        const float4* F = reinterpret_cast<const float4*>(fb_local + 8 * b);
        const float4* S = reinterpret_cast<const float4*>(sb + 8 * b);
        const float4 n0 = upd4(F[0], c0, __ldg(S)), n1 = upd4(F[1], c1, __ldg(S + 1));
        if (MM) {
            float* pf = (float*)ncclGetLsaMultimemPointer(wf, off, dc);
            mm_st4(pf, n0);
            mm_st4(pf + 4, n1);
        } else {
            for (int p = 0; p < nr; ++p) {
                float4* pf = (float4*)ncclGetLsaPointer(wf, off, p);
                pf[0] = n0;
                pf[1] = n1;
            }
        }
    }
    {
        ncclLsaBarrierSession<ncclCoopCta> bar(ncclCoopCta(), dc, ncclTeamTagLsa(), blockIdx.x, MM);
        bar.sync(ncclCoopCta(), cuda::memory_order_acq_rel);
    }
    // CTA k of every rank has read its bricks of every c: re-zero those bricks locally
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
