// k_update_block.cu — unit test of the ISD block update (lmk::k_update with a brick block
// and zero_to, the one-launch form used after ncclReduceScatter): inside the block
// f <- f*c/s where c > 0 and s > 0 (reading S9) and c <- 0; outside the block but
// below zero_to only c <- 0; beyond zero_to nothing changes. Exit 0 and "ok" on success.
#include <cstdio>
#include <cstdlib>
#include <vector>

#include "lmosem_kernels.cuh"

static unsigned lcg(unsigned& x) { return x = x * 1664525u + 1013904223u; }

int main() {
    const int64_t nb = 1000, nbf = 8 * nb;
    const int64_t cases[][3] = {{0, nb, nb}, {250, 500, nb}, {0, 125, nb}, {875, 1000, nb},
                                {900, 900, nb}, {300, 700, 800}, {990, 995, 1000}};
    lmk::GridGeom g{};  // f_row is null: the geometry is not read
    lmk::BrickIt it{10, 10, 10, nb};
    float *df, *dc, *ds;
    cudaMalloc(&df, 4 * nbf);
    cudaMalloc(&dc, 4 * nbf);
    cudaMalloc(&ds, 4 * nbf);
    unsigned x = 12345;
    int bad = 0;
    for (const auto& cs : cases) {
        const int64_t b0 = cs[0], b1 = cs[1], zt = cs[2];
        std::vector<float> f(nbf), c(nbf), s(nbf), fo(nbf), co(nbf);
        for (int64_t i = 0; i < nbf; ++i) {
            f[i] = 0.5f + (lcg(x) >> 8) * (1.0f / 16777216.0f);
            c[i] = (lcg(x) % 5 == 0) ? 0.0f : (lcg(x) >> 8) * (1.0f / 16777216.0f);
            s[i] = (lcg(x) % 7 == 0) ? 0.0f : 0.2f + (lcg(x) >> 8) * (1.0f / 16777216.0f);
        }
        cudaMemcpy(df, f.data(), 4 * nbf, cudaMemcpyHostToDevice);
        cudaMemcpy(dc, c.data(), 4 * nbf, cudaMemcpyHostToDevice);
        cudaMemcpy(ds, s.data(), 4 * nbf, cudaMemcpyHostToDevice);
        lmk::k_update<<<7, 256>>>(df, dc, ds, nullptr, g, it, b0, b1, zt);
        if (cudaDeviceSynchronize() != cudaSuccess) {
            std::printf("launch failed\n");
            return 1;
        }
        cudaMemcpy(fo.data(), df, 4 * nbf, cudaMemcpyDeviceToHost);
        cudaMemcpy(co.data(), dc, 4 * nbf, cudaMemcpyDeviceToHost);
        for (int64_t i = 0; i < nbf; ++i) {
            const int64_t b = i / 8;
            const bool in = b >= b0 && b < b1, zero = b < zt;
            const float q = c[i] / s[i];  // IEEE single division, as __fdiv_rn
            const float fe = in && c[i] > 0.0f && s[i] > 0.0f ? f[i] * q : f[i];
            const float ce = (in || zero) ? 0.0f : c[i];
            if (fo[i] != fe || co[i] != ce) {
                if (bad++ < 5)
                    std::printf("case [%lld,%lld) zero_to %lld: element %lld f %g (want %g) c %g (want %g)\n",
                                (long long)b0, (long long)b1, (long long)zt, (long long)i, fo[i], fe, co[i], ce);
            }
        }
    }
    cudaFree(df);
    cudaFree(dc);
    cudaFree(ds);
    if (bad) {
        std::printf("%d mismatches\n", bad);
        return 1;
    }
    std::printf("ok\n");
    return 0;
}
