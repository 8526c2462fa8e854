// combine_emu.cu — the fused ISD combine body (lmk::combine_fused_body, §8(f) NEXT-1) with P
// emulated ranks on ONE GPU: one kernel of P x ctas CTAs, CTA (r, k) plays CTA k of rank r;
// every rank has its own c, brick f and norm buffers; the team barrier is a global-memory
// counter per k (all CTAs are co-resident). Checks, bitwise against the host, that every
// rank ends with f_j <- f_j * (sum_p c_p,j) / s_j where the sum > 0 and s_j > 0 (the sum
// taken over p = 0..P-1 in order, as the peer-pointer team does), and with c = 0 everywhere.
// Multi-rank logic only: NCCL's LSA barrier, windows and multimem are not exercised.
#include <cstdio>
#include <vector>

#include "lmosem_kernels.cuh"

struct EmuTeam {
    float* const* c;  // c of every rank
    float* const* f;  // brick f of every rank
    unsigned* bar;    // one arrival counter per CTA index k
    int r, P;
    unsigned epoch;
    __device__ __forceinline__ void sync(int k) {
        ++epoch;
        __syncthreads();
        if (threadIdx.x == 0) {
            __threadfence();
            atomicAdd(bar + k, 1u);
            while (*(volatile unsigned*)(bar + k) < epoch * (unsigned)P) {
            }
            __threadfence();
        }
        __syncthreads();
    }
    __device__ __forceinline__ int rank() const { return r; }
    __device__ __forceinline__ int size() const { return P; }
    __device__ __forceinline__ void sum_c(size_t off, float4& c0, float4& c1) {
        c0 = make_float4(0.f, 0.f, 0.f, 0.f);
        c1 = c0;
        for (int p = 0; p < P; ++p) {
            const float4* pc = reinterpret_cast<const float4*>(reinterpret_cast<const char*>(c[p]) + off);
            c0 = lmk::add4(c0, __ldcg(pc));
            c1 = lmk::add4(c1, __ldcg(pc + 1));
        }
    }
    __device__ __forceinline__ void sum_c2(size_t oa, size_t ob, float4& a0, float4& a1, float4& b0, float4& b1) {
        sum_c(oa, a0, a1);
        sum_c(ob, b0, b1);
    }
    __device__ __forceinline__ void store_f(size_t off, float4 n0, float4 n1) {
        for (int p = 0; p < P; ++p) {
            float4* pf = reinterpret_cast<float4*>(reinterpret_cast<char*>(f[p]) + off);
            __stcg(pf, n0);
            __stcg(pf + 1, n1);
        }
    }
};

__global__ void __launch_bounds__(256) k_emu(float* const* c, float* const* f, float* const* s, unsigned* bar, int P,
                                             int ctas, int64_t chunk, int64_t nb) {
    const int r = blockIdx.x / ctas, k = blockIdx.x % ctas;
    EmuTeam team{c, f, bar, r, P, 0u};
    lmk::combine_fused_body(team, k, ctas, s[r], c[r], f[r], chunk, nb, lmk::BrickIt{});
}

static unsigned lcg(unsigned& x) { return x = x * 1664525u + 1013904223u; }
static float u01(unsigned& x) { return (lcg(x) >> 8) * (1.0f / 16777216.0f); }

int main() {
    int bad = 0;
    unsigned x = 777;
    const int64_t nbs[] = {1, 7, 1000, 4099};
    for (int P : {1, 2, 3, 4, 8}) {
        for (int64_t nb : nbs) {
            const int64_t nb_alloc = (nb + P - 1) / P * P, chunk = nb_alloc / P, nbf = 8 * nb_alloc;
            const int ctas = 4 * 148 / P;  // all P x ctas CTAs co-resident (4 per SM), as in production
            // host images per rank: c (partial error images), brick f (identical replicas), s
            std::vector<std::vector<float>> c(P, std::vector<float>(nbf)), f(P), s(P);
            std::vector<float> f0(nbf), s0(nbf);
            for (int64_t i = 0; i < nbf; ++i) {
                f0[i] = 0.5f + u01(x);
                s0[i] = (lcg(x) % 9 == 0) ? 0.0f : 0.2f + u01(x);
            }
            for (int p = 0; p < P; ++p) {
                for (int64_t i = 0; i < nbf; ++i) c[p][i] = (lcg(x) % 6 == 0) ? 0.0f : u01(x);
                f[p] = f0;
                s[p] = s0;
            }
            std::vector<float*> dc(P), df(P), ds(P);
            for (int p = 0; p < P; ++p) {
                cudaMalloc(&dc[p], 4 * nbf);
                cudaMalloc(&df[p], 4 * nbf);
                cudaMalloc(&ds[p], 4 * nbf);
                cudaMemcpy(dc[p], c[p].data(), 4 * nbf, cudaMemcpyHostToDevice);
                cudaMemcpy(df[p], f[p].data(), 4 * nbf, cudaMemcpyHostToDevice);
                cudaMemcpy(ds[p], s[p].data(), 4 * nbf, cudaMemcpyHostToDevice);
            }
            float **pc, **pf, **ps;
            unsigned* bar;
            cudaMalloc(&pc, sizeof(float*) * P);
            cudaMalloc(&pf, sizeof(float*) * P);
            cudaMalloc(&ps, sizeof(float*) * P);
            cudaMalloc(&bar, sizeof(unsigned) * ctas);
            cudaMemset(bar, 0, sizeof(unsigned) * ctas);
            cudaMemcpy(pc, dc.data(), sizeof(float*) * P, cudaMemcpyHostToDevice);
            cudaMemcpy(pf, df.data(), sizeof(float*) * P, cudaMemcpyHostToDevice);
            cudaMemcpy(ps, ds.data(), sizeof(float*) * P, cudaMemcpyHostToDevice);
            k_emu<<<P * ctas, 256>>>(pc, pf, ps, bar, P, ctas, chunk, nb);
            if (cudaDeviceSynchronize() != cudaSuccess) {
                std::printf("launch failed (P=%d nb=%lld)\n", P, (long long)nb);
                return 1;
            }
            // expected: real bricks [0, nb) updated with the rank-ordered sum; padding
            // bricks [nb, nb_alloc) untouched in f; c zero on [0, nb) of every rank
            std::vector<float> fe(nbf);
            for (int64_t i = 0; i < nbf; ++i) {
                if (i >= 8 * nb) {
                    fe[i] = f0[i];
                    continue;
                }
                float sum = 0.0f;
                for (int p = 0; p < P; ++p) sum += c[p][i];
                const float q = sum / s0[i];
                fe[i] = (sum > 0.0f && s0[i] > 0.0f) ? f0[i] * q : f0[i];
            }
            for (int p = 0; p < P; ++p) {
                std::vector<float> fo(nbf), co(nbf);
                cudaMemcpy(fo.data(), df[p], 4 * nbf, cudaMemcpyDeviceToHost);
                cudaMemcpy(co.data(), dc[p], 4 * nbf, cudaMemcpyDeviceToHost);
                for (int64_t i = 0; i < nbf; ++i) {
                    const float ce = i < 8 * nb ? 0.0f : c[p][i];
                    if (fo[i] != fe[i] || co[i] != ce) {
                        if (bad++ < 8)
                            std::printf("P=%d nb=%lld rank %d elem %lld: f %g (want %g) c %g (want %g)\n", P,
                                        (long long)nb, p, (long long)i, fo[i], fe[i], co[i], ce);
                    }
                }
                cudaFree(dc[p]);
                cudaFree(df[p]);
                cudaFree(ds[p]);
            }
            cudaFree(pc);
            cudaFree(pf);
            cudaFree(ps);
            cudaFree(bar);
        }
    }
    if (bad) {
        std::printf("%d mismatches\n", bad);
        return 1;
    }
    std::printf("ok\n");
    return 0;
}
