// request_probe.cu — probe: does the L1->L2 path limit 32-byte *sectors* or *requests*
// (one request = the sectors of one 128-byte line a warp instruction touches)?
// Every warp instruction touches 16 sectors with 2 lanes per sector (the projection's
// ~2 path pieces per sector), spread over 16 / k random 128-byte lines of k sectors each
// (k = 1, 2, 4), on an L2-resident buffer of V floats (C2: 25.2 MB). Reports sectors/s
// and requests/s for LSU gathers (ld.global.nc.f32), REDs (red.global.add.f32) and a
// gather+RED mix of the same addresses.
// Standalone: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o request_probe request_probe.cu
#include <cuda_runtime.h>
#include <stdint.h>
#include <stdio.h>

__device__ __forceinline__ uint32_t hash32(uint32_t x) {
    x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16;
    return x;
}

// OP 0: gather, 1: RED, 2: gather then RED of the same float
template <int OP, int K>
__global__ void __launch_bounds__(256) k(float* __restrict__ buf, uint32_t nlines, int ops, float* sink) {
    const int lane = threadIdx.x & 31;
    const uint32_t warp = (blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    // lane -> (line slot, sector in line, lane in sector): 2 lanes per sector, K sectors per line
    const int sec_in_warp = lane >> 1;             // 0..15
    const int line_slot = sec_in_warp / K;         // 0..16/K-1
    const int sec_in_line = sec_in_warp % K;       // 0..K-1
    const int off = sec_in_line * 8 + (lane & 1) * 3;
    float acc = 0.f;
    for (int it = 0; it < ops; ++it) {
        const uint32_t key = (warp * 16u + (uint32_t)line_slot) * 0x9E3779B9u + (uint32_t)it * 0x85EBCA6Bu;
        const uint32_t ln = (uint32_t)(((uint64_t)hash32(key) * (nlines - 1)) >> 32);
        // K < 4: a random K-sector-aligned group inside the line
        const uint32_t grp = (hash32(key ^ 0xABCDu) % (4 / K)) * K;
        float* p = buf + 32ull * ln + grp * 8 + off;
        if (OP == 0 || OP == 2) acc += __ldg(p);
        if (OP == 1) atomicAdd(p, 1.0f);
        if (OP == 2) atomicAdd(p, acc * 1e-30f);
    }
    if (acc == 12345.f) sink[0] = acc;
}

template <int OP, int K>
float run(float* buf, uint32_t nlines, int grid, int ops, float* sink) {
    cudaEvent_t a, b;
    cudaEventCreate(&a);
    cudaEventCreate(&b);
    k<OP, K><<<grid, 256>>>(buf, nlines, ops, sink);
    cudaEventRecord(a);
    for (int r = 0; r < 5; ++r) k<OP, K><<<grid, 256>>>(buf, nlines, ops, sink);
    cudaEventRecord(b);
    cudaEventSynchronize(b);
    float ms;
    cudaEventElapsedTime(&ms, a, b);
    return ms / 5;
}

template <int OP, int K>
void report(const char* name, float* buf, uint32_t nlines, int grid, int ops, float* sink) {
    const float ms = run<OP, K>(buf, nlines, grid, ops, sink);
    const double warps = (double)grid * 8, instr = warps * ops * (OP == 2 ? 2 : 1);
    const double sectors = instr * 16, requests = instr * (16 / K);
    printf("%-8s k=%d sectors/line: %.3e sectors/s  %.3e requests/s  (%.3f ms)\n", name, K, sectors / (ms * 1e-3),
           requests / (ms * 1e-3), ms);
}

int main() {
    const uint64_t V = 6735344ull * 8 / 8;  // C2 padded brick image (floats)
    const uint32_t nlines = (uint32_t)(V / 32);
    float *buf, *sink;
    cudaMalloc(&buf, V * 4);
    cudaMalloc(&sink, 4);
    cudaMemset(buf, 0, V * 4);
    int sms;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    const int grid = sms * 8, ops = 2000;
    report<0, 1>("gather", buf, nlines, grid, ops, sink);
    report<0, 2>("gather", buf, nlines, grid, ops, sink);
    report<0, 4>("gather", buf, nlines, grid, ops, sink);
    report<1, 1>("red", buf, nlines, grid, ops, sink);
    report<1, 2>("red", buf, nlines, grid, ops, sink);
    report<1, 4>("red", buf, nlines, grid, ops, sink);
    report<2, 1>("pair", buf, nlines, grid, ops, sink);
    report<2, 2>("pair", buf, nlines, grid, ops, sink);
    report<2, 4>("pair", buf, nlines, grid, ops, sink);
    cudaError_t e = cudaDeviceSynchronize();
    printf("%s\n", cudaGetErrorString(e));
    return 0;
}
