// l2peak.cu — microbenchmarks for the L2 roofline denominators (include/l2peak.h).
#include <cuda_runtime.h>
#include <stdint.h>

#include "l2peak.h"

#define L2PEAK_API extern "C" __attribute__((visibility("default")))

namespace {

__device__ __forceinline__ uint32_t hash32(uint32_t x) {
    x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16;
    return x;
}

template <int MODE>
__global__ void __launch_bounds__(256) k_l2(float* __restrict__ buf, const float* __restrict__ src, uint32_t n,
                                            int ops, float* __restrict__ sink) {
    const uint32_t tid = blockIdx.x * blockDim.x + threadIdx.x;
    const int lane = threadIdx.x & 31;
    float acc = 0.f;
#pragma unroll 4
    for (int it = 0; it < ops; ++it) {
        uint32_t h = hash32(tid * 0x9E3779B9u + (uint32_t)it * 0x85EBCA6Bu);
        uint32_t j;
        if (MODE == L2PEAK_PAIR_WARP32 || MODE == L2PEAK_LDG_WARP32 || MODE == L2PEAK_RED_WARP32) {
            uint32_t g = hash32((tid >> 5) * 0x9E3779B9u + (uint32_t)it * 0x85EBCA6Bu);
            j = ((uint32_t)(((uint64_t)g * (n - 32)) >> 32) & ~31u) + lane;
        } else if (MODE == L2PEAK_RED_RUN8 || MODE == L2PEAK_PAIR_RUN8) {
            uint32_t g = hash32((tid >> 3) * 0x9E3779B9u + (uint32_t)it * 0x85EBCA6Bu);
            j = (uint32_t)(((uint64_t)g * (n - 8)) >> 32) + (lane & 7);
        } else {
            j = (uint32_t)(((uint64_t)h * n) >> 32);
        }
        if (MODE == L2PEAK_LDG_RANDOM || MODE == L2PEAK_PAIR_RANDOM || MODE == L2PEAK_PAIR_RUN8 ||
            MODE == L2PEAK_PAIR_WARP32 || MODE == L2PEAK_LDG_WARP32)
            acc += __ldg(src + j);
        if (MODE != L2PEAK_LDG_RANDOM && MODE != L2PEAK_LDG_WARP32) atomicAdd(buf + j, 1.0f + acc * 0.0f);
    }
    if (acc == 12345.678f) sink[0] = acc;  // keeps the gathers alive
}

// STREAM5: the update kernel's access pattern, streamed: read a, b, c, write a, b (float4),
// a grid-stride pass over n floats per array, `ops` passes (the arrays stay L2-resident
// when 3 * 4 * n bytes fit).
__global__ void __launch_bounds__(256) k_stream5(float4* __restrict__ a, float4* __restrict__ b,
                                                 const float4* __restrict__ c, uint32_t n4, int ops) {
    for (int it = 0; it < ops; ++it)
        for (uint32_t i = blockIdx.x * blockDim.x + threadIdx.x; i < n4; i += gridDim.x * blockDim.x) {
            float4 x = a[i], y = b[i];
            const float4 z = c[i];
            x.x = x.x * y.x + z.x; x.y = x.y * y.y + z.y; x.z = x.z * y.z + z.z; x.w = x.w * y.w + z.w;
            a[i] = x;
            b[i] = make_float4(0.f, 0.f, 0.f, 0.f);
        }
}

template <int MODE>
cudaError_t launch(float* buf, const float* src, uint32_t n, int ops, float* sink, int grid) {
    k_l2<MODE><<<grid, 256>>>(buf, src, n, ops, sink);
    return cudaGetLastError();
}

cudaError_t launch_mode(int mode, float* buf, const float* src, uint32_t n, int ops, float* sink, int grid) {
    switch (mode) {
        case L2PEAK_RED_RANDOM: return launch<L2PEAK_RED_RANDOM>(buf, src, n, ops, sink, grid);
        case L2PEAK_LDG_RANDOM: return launch<L2PEAK_LDG_RANDOM>(buf, src, n, ops, sink, grid);
        case L2PEAK_PAIR_RANDOM: return launch<L2PEAK_PAIR_RANDOM>(buf, src, n, ops, sink, grid);
        case L2PEAK_RED_RUN8: return launch<L2PEAK_RED_RUN8>(buf, src, n, ops, sink, grid);
        case L2PEAK_PAIR_RUN8: return launch<L2PEAK_PAIR_RUN8>(buf, src, n, ops, sink, grid);
        case L2PEAK_PAIR_WARP32: return launch<L2PEAK_PAIR_WARP32>(buf, src, n, ops, sink, grid);
        case L2PEAK_LDG_WARP32: return launch<L2PEAK_LDG_WARP32>(buf, src, n, ops, sink, grid);
        case L2PEAK_RED_WARP32: return launch<L2PEAK_RED_WARP32>(buf, src, n, ops, sink, grid);
        case L2PEAK_STREAM5:
            k_stream5<<<grid, 256>>>(reinterpret_cast<float4*>(buf), const_cast<float4*>(reinterpret_cast<const float4*>(src)),
                                     reinterpret_cast<const float4*>(sink), n / 4, ops);
            return cudaGetLastError();
    }
    return cudaErrorInvalidValue;
}

}  // namespace

L2PEAK_API int l2peak_run(int mode, int64_t n_floats, int32_t ops_per_thread, float* ms, double* ops) {
    if (mode < 0 || mode > L2PEAK_RED_WARP32 || n_floats < 64 || n_floats >= (int64_t(1) << 32) || ops_per_thread <= 0 || !ms || !ops)
        return -1;
    int dev = 0, sms = 0, per_sm = 0;
    if (cudaGetDevice(&dev) != cudaSuccess) return -1;
    if (cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev) != cudaSuccess) return -1;
    cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k_l2<L2PEAK_PAIR_RANDOM>, 256, 0);
    if (per_sm < 1) per_sm = 1;
    const int grid = sms * per_sm;
    float *buf = nullptr, *src = nullptr, *sink = nullptr;
    cudaEvent_t e0 = nullptr, e1 = nullptr;
    int rc = -1;
    if (cudaMalloc(&buf, sizeof(float) * n_floats) != cudaSuccess) goto done;
    if (cudaMalloc(&src, sizeof(float) * n_floats) != cudaSuccess) goto done;
    if (cudaMalloc(&sink, sizeof(float) * (mode == L2PEAK_STREAM5 ? n_floats : 1)) != cudaSuccess) goto done;
    if (mode == L2PEAK_STREAM5) cudaMemset(sink, 0, sizeof(float) * n_floats);
    cudaMemset(buf, 0, sizeof(float) * n_floats);
    cudaMemset(src, 0, sizeof(float) * n_floats);
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    if (launch_mode(mode, buf, src, (uint32_t)n_floats, ops_per_thread, sink, grid) != cudaSuccess) goto done;
    cudaEventRecord(e0);
    if (launch_mode(mode, buf, src, (uint32_t)n_floats, ops_per_thread, sink, grid) != cudaSuccess) goto done;
    cudaEventRecord(e1);
    if (cudaEventSynchronize(e1) != cudaSuccess) goto done;
    cudaEventElapsedTime(ms, e0, e1);
    *ops = mode == L2PEAK_STREAM5 ? (double)(n_floats / 4 * 4) * ops_per_thread : (double)grid * 256.0 * ops_per_thread;
    rc = 0;
done:
    if (e0) cudaEventDestroy(e0);
    if (e1) cudaEventDestroy(e1);
    cudaFree(buf);
    cudaFree(src);
    cudaFree(sink);
    return rc;
}
