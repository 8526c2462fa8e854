/* abi_consumer.c — a plain C99 user of the LM-OSEM C ABI (include/lmosem.h): no Python, no
 * torch; device memory from the CUDA runtime. Proves the boundary is usable on its own
 * (tests/test_abi_c.py compiles it on CPU and runs it on the GPU against the oracle).
 *
 *   abi_consumer nx ny nz vx vy vz events.bin norm.bin n_events n_subsets iters out.bin
 *
 * events.bin: n_events lmosem_event records; norm.bin: V float32. Runs
 * lmosem_reconstruct (device buffers) and lmosem_reconstruct_host (host buffers) over
 * n_subsets equal contiguous subsets from f0 = 1 and writes both results (2 x V float32)
 * to out.bin. Also checks argument errors. Exit 0 on success, else prints the failure. */
#include <cuda_runtime_api.h>
#include <stdio.h>
#include <stdlib.h>
#include <string.h>

#include "lmosem.h"

#define CHECK(call)                                                                      \
    do {                                                                                 \
        lmosem_status st_ = (call);                                                      \
        if (st_ != LMOSEM_OK) {                                                          \
            fprintf(stderr, "%s:%d %s -> %d (%s)\n", __FILE__, __LINE__, #call, (int)st_, \
                    lmosem_last_error(ctx));                                             \
            return 1;                                                                    \
        }                                                                                \
    } while (0)

#define CUDA(call)                                                                          \
    do {                                                                                    \
        cudaError_t e_ = (call);                                                            \
        if (e_ != cudaSuccess) {                                                            \
            fprintf(stderr, "%s:%d %s -> %s\n", __FILE__, __LINE__, #call, cudaGetErrorString(e_)); \
            return 1;                                                                       \
        }                                                                                   \
    } while (0)

static void* read_file(const char* path, size_t bytes) {
    FILE* fh = fopen(path, "rb");
    void* p = malloc(bytes ? bytes : 1);
    if (!fh || !p || fread(p, 1, bytes, fh) != bytes) {
        if (fh) fclose(fh);
        free(p);
        return NULL;
    }
    fclose(fh);
    return p;
}

int main(int argc, char** argv) {
    lmosem_ctx* ctx = NULL;
    if (argc != 13) {
        fprintf(stderr, "usage: %s nx ny nz vx vy vz events.bin norm.bin n_events n_subsets iters out.bin\n", argv[0]);
        return 2;
    }
    const int32_t dims[3] = {atoi(argv[1]), atoi(argv[2]), atoi(argv[3])};
    const double vox[3] = {atof(argv[4]), atof(argv[5]), atof(argv[6])};
    const int64_t n = atoll(argv[9]);
    const int32_t L = atoi(argv[10]), iters = atoi(argv[11]);
    const int64_t V = (int64_t)dims[0] * dims[1] * dims[2];
    lmosem_event* ev = (lmosem_event*)read_file(argv[7], sizeof(lmosem_event) * (size_t)n);
    float* norm = (float*)read_file(argv[8], sizeof(float) * (size_t)V);
    if (!ev || !norm || L < 1) {
        fprintf(stderr, "cannot read inputs\n");
        return 2;
    }
    printf("%s\n", lmosem_version());

    /* argument errors: nothing is created, the status says why */
    {
        const int32_t bad[3] = {0, dims[1], dims[2]};
        lmosem_ctx* none = (lmosem_ctx*)1;
        if (lmosem_init(&none, bad, vox, norm, NULL) != LMOSEM_EINVAL || none != NULL) {
            fprintf(stderr, "zero extent not rejected\n");
            return 1;
        }
        int64_t b, e;
        if (lmosem_block_range(10, 3, 2, &b, &e) != LMOSEM_EINVAL) return 1;
        CHECK(lmosem_block_range(10, 1, 3, &b, &e));
        if (b != 3 || e != 6) return 1;
    }

    int64_t* off = (int64_t*)malloc(sizeof(int64_t) * (size_t)(L + 1));
    for (int32_t l = 0; l <= L; ++l) off[l] = (n * l) / L;

    CHECK(lmosem_init(&ctx, dims, vox, norm, NULL)); /* host norm: copied */
    lmosem_event* d_ev = NULL;
    float* d_f = NULL;
    CUDA(cudaMalloc((void**)&d_ev, sizeof(lmosem_event) * (size_t)(n ? n : 1)));
    CUDA(cudaMalloc((void**)&d_f, sizeof(float) * (size_t)V));
    CUDA(cudaMemcpy(d_ev, ev, sizeof(lmosem_event) * (size_t)n, cudaMemcpyHostToDevice));
    float* f = (float*)malloc(sizeof(float) * (size_t)V * 2);
    for (int64_t j = 0; j < V; ++j) f[j] = 1.0f;
    CUDA(cudaMemcpy(d_f, f, sizeof(float) * (size_t)V, cudaMemcpyHostToDevice));

    /* device buffers, stream-ordered: synchronize before reading f */
    CHECK(lmosem_reconstruct(ctx, d_ev, off, L, iters, d_f));
    CHECK(lmosem_synchronize(ctx));
    CUDA(cudaMemcpy(f, d_f, sizeof(float) * (size_t)V, cudaMemcpyDeviceToHost));

    /* pageable host memory is not a device buffer: EINVAL, context still usable */
    if (lmosem_subset_step(ctx, ev, n, d_f) != (n ? LMOSEM_EINVAL : LMOSEM_OK)) {
        fprintf(stderr, "pageable events not rejected\n");
        return 1;
    }

    /* host buffers (synchronous; pinned memory overlaps the copies) */
    lmosem_event* h_ev = NULL;
    float* h_f = NULL;
    CUDA(cudaMallocHost((void**)&h_ev, sizeof(lmosem_event) * (size_t)(n ? n : 1)));
    CUDA(cudaMallocHost((void**)&h_f, sizeof(float) * (size_t)V));
    memcpy(h_ev, ev, sizeof(lmosem_event) * (size_t)n);
    for (int64_t j = 0; j < V; ++j) h_f[j] = 1.0f;
    CHECK(lmosem_reconstruct_host(ctx, h_ev, off, L, iters, h_f));
    memcpy(f + V, h_f, sizeof(float) * (size_t)V);

    lmosem_stats st;
    CHECK(lmosem_get_stats(ctx, &st));
    printf("subsets %lld launches %lld events %lld\n", (long long)st.subsets, (long long)st.launches,
           (long long)st.events);
    CHECK(lmosem_destroy(ctx));
    ctx = NULL;

    FILE* out = fopen(argv[12], "wb");
    if (!out || fwrite(f, sizeof(float), (size_t)V * 2, out) != (size_t)V * 2) return 1;
    fclose(out);
    cudaFree(d_ev);
    cudaFree(d_f);
    cudaFreeHost(h_ev);
    cudaFreeHost(h_f);
    free(ev);
    free(norm);
    free(off);
    free(f);
    printf("ok\n");
    return 0;
}
