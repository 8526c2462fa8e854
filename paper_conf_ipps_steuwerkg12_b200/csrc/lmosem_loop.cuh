// lmosem_loop.cuh — kernels of the loopback transport (include/lmosem.h, "Emulated world"):
// P contexts of one process on ONE GPU stand in for P ranks, so the multi-GPU combine of
// the subset iteration (Listing 3 l.6 and l.15-16: the per-GPU
// error images are added, step 2 runs on the sum, f is replicated again) runs through the
// same subset_iteration code as the NCCL build and can be checked against the oracle with
// one GPU. The collectives keep NCCL's semantics; each rank's part is one kernel that reads
// the other ranks' buffers directly (same device), ordered by events behind a host barrier
// (lmosem.cu). The fused combine (§8(f) NEXT-1) runs the same combine_fused_body as
// k_combine_fused, with a team whose barrier is a device counter per CTA index.
#pragma once
#include <cuda/atomic>

#include "lmosem_kernels.cuh"

namespace lmk {

constexpr int kLoopMax = 16;  // largest emulated world

struct LoopSrc {
    const float* p[kLoopMax];
    int64_t off[kLoopMax + 1];  // all-gather: region q of the destination is [off[q], off[q+1])
};

// reduce: dst[i] = sum over q = 0..P-1 (in rank order) of src.p[q][i], i < count
__global__ void __launch_bounds__(256) k_loop_sum(LoopSrc src, float* __restrict__ dst, int64_t count, int P) {
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < count; i += (int64_t)gridDim.x * blockDim.x) {
        float a = src.p[0][i];
        for (int q = 1; q < P; ++q) a += src.p[q][i];
        dst[i] = a;
    }
}

// gather: dst[off[q] + i] = src.p[q][i] for every q != self (blockIdx.y = q), i < off[q+1] - off[q]
__global__ void __launch_bounds__(256) k_loop_gather(LoopSrc src, float* __restrict__ dst, int self) {
    const int q = blockIdx.y;
    if (q == self) return;  // in place: this rank's own region is already in dst
    const int64_t n = src.off[q + 1] - src.off[q];
    const float* s = src.p[q];
    float* d = dst + src.off[q];
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x)
        d[i] = s[i];
}

// ------------------------------------------------------------ emulated fused combine team
struct LoopImages {
    float* c[kLoopMax];         // error image (bricks) of every rank
    float* fb[kLoopMax];        // brick f of every rank
    const float* s[kLoopMax];   // norm (bricks) of every rank
};

// The team of combine_fused_body for P emulated ranks: CTA (r, k) of one cooperative launch
// plays CTA k of rank r; sync(k) is a barrier of the P CTAs with index k (device counter,
// release/acquire), like the LSA barrier of CTA k across the ranks in the NCCL team.
struct LoopTeam {
    const LoopImages* im;
    unsigned* bar;  // one arrival counter per CTA index k, zeroed before the launch
    int r, P;
    unsigned epoch;
    __device__ __forceinline__ void sync(int k) {
        ++epoch;
        __syncthreads();
        if (threadIdx.x == 0) {
            cuda::atomic_ref<unsigned, cuda::thread_scope_device> a(bar[k]);
            a.fetch_add(1u, cuda::memory_order_release);
            while (a.load(cuda::memory_order_acquire) < epoch * (unsigned)P) __nanosleep(64);
        }
        __syncthreads();
    }
    __device__ __forceinline__ int rank() const { return r; }
    __device__ __forceinline__ int size() const { return P; }
    __device__ __forceinline__ void sum_c(size_t off, float4& c0, float4& c1) {
        c0 = make_float4(0.f, 0.f, 0.f, 0.f);
        c1 = c0;
        for (int p = 0; p < P; ++p) {
            const float4* pc = reinterpret_cast<const float4*>(reinterpret_cast<const char*>(im->c[p]) + off);
            c0 = add4(c0, __ldcg(pc));
            c1 = add4(c1, __ldcg(pc + 1));
        }
    }
    __device__ __forceinline__ void sum_c2(size_t oa, size_t ob, float4& a0, float4& a1, float4& b0, float4& b1) {
        sum_c(oa, a0, a1);
        sum_c(ob, b0, b1);
    }
    __device__ __forceinline__ void store_f(size_t off, float4 n0, float4 n1) {
        for (int p = 0; p < P; ++p) {
            float4* pf = reinterpret_cast<float4*>(reinterpret_cast<char*>(im->fb[p]) + off);
            __stcg(pf, n0);
            __stcg(pf + 1, n1);
        }
    }
};

// One cooperative launch of P * ctas CTAs (all co-resident, so the spin barrier is safe).
__global__ void __launch_bounds__(256) k_combine_loop(LoopImages im, unsigned* bar, int P, int ctas, int64_t chunk,
                                                      int64_t nb, BrickIt it) {
    const int r = blockIdx.x / ctas, k = blockIdx.x % ctas;
    LoopTeam team{&im, bar, r, P, 0u};
    combine_fused_body(team, k, ctas, im.s[r], im.c[r], im.fb[r], chunk, nb, it);
}

}  // namespace lmk
