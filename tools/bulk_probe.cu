// bulk_probe.cu — probe: is the projection's scattered-sector rate an SM (LSU / L1 miss
// path) limit or an L2 limit?  Compares, on an L2-resident V-float buffer, the 32-byte
// sector rate of
//   0  LSU red.global.add.f32, 2 lanes per sector (the projection's ~2 pieces / sector)
//   1  LSU red.global.add.v4.f32 (16 B per lane), 2 lanes per sector
//   2  LSU 2 x red.global.add.v4.f32 by one lane (one lane per sector)
//   3  TMA bulk reduce cp.reduce.async.bulk .add.f32 of 32 B per op (one op per sector)
//   4  TMA bulk reduce of 64 B per op (two sectors)
//   5  LSU gather ld.global.f32, 2 lanes per sector
//   6  TMA bulk copy global -> smem of 32 B per op (gather of one sector)
//   7  LSU gather ld.global.v8.f32 (one lane per sector)
// Standalone: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o bulk_probe bulk_probe.cu
#include <cuda_runtime.h>
#include <stdint.h>
#include <stdio.h>

__device__ __forceinline__ uint32_t hash32(uint32_t x) {
    x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16;
    return x;
}

template <int MODE>
__global__ void __launch_bounds__(256) k(float* __restrict__ buf, uint32_t nsec, int ops, float* sink) {
    __shared__ __align__(128) float slot[256 * 16];
    __shared__ __align__(8) unsigned long long bar[8];
    const uint32_t tid = blockIdx.x * blockDim.x + threadIdx.x;
    const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
    for (int q = 0; q < 16; ++q) slot[threadIdx.x * 16 + q] = 1.0f;
    if (lane == 0) asm volatile("mbarrier.init.shared.b64 [%0], 1;" ::"r"((unsigned)__cvta_generic_to_shared(&bar[w])));
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
    __syncthreads();
    const unsigned my_s = (unsigned)__cvta_generic_to_shared(&slot[threadIdx.x * 16]);
    const unsigned bar_s = (unsigned)__cvta_generic_to_shared(&bar[w]);
    float acc = 0.f;
    unsigned phase = 0;
    for (int it = 0; it < ops; ++it) {
        // sector index: pairs of lanes share a sector for the 2-lanes-per-sector modes
        const bool pairs = (MODE == 0 || MODE == 1 || MODE == 5);
        const uint32_t key = pairs ? (tid >> 1) : tid;
        const uint32_t s = (uint32_t)(((uint64_t)hash32(key * 0x9E3779B9u + (uint32_t)it * 0x85EBCA6Bu) * (nsec - 2)) >> 32);
        float* sec = buf + 8ull * s;
        if (MODE == 0) {
            atomicAdd(sec + (lane & 1) * 3, 1.0f);
        } else if (MODE == 1) {
            float* p = sec + (lane & 1) * 4;
            asm volatile("red.global.add.v4.f32 [%0], {%1, %1, %1, %1};" ::"l"(p), "f"(1.0f) : "memory");
        } else if (MODE == 2) {
            asm volatile("red.global.add.v4.f32 [%0], {%1, %1, %1, %1};" ::"l"(sec), "f"(1.0f) : "memory");
            asm volatile("red.global.add.v4.f32 [%0], {%1, %1, %1, %1};" ::"l"(sec + 4), "f"(1.0f) : "memory");
        } else if (MODE == 3 || MODE == 4) {
            asm volatile("cp.reduce.async.bulk.global.shared::cta.bulk_group.add.f32 [%0], [%1], %2;" ::"l"(sec),
                         "r"(my_s), "n"(MODE == 3 ? 32 : 64)
                         : "memory");
            asm volatile("cp.async.bulk.commit_group;" ::: "memory");
            if ((it & 7) == 7) asm volatile("cp.async.bulk.wait_group.read 4;" ::: "memory");
        } else if (MODE == 5) {
            acc += __ldg(sec + (lane & 1) * 3);
        } else if (MODE == 6) {
            // batches of 8 sectors per lane per mbarrier phase: lane 0 expects the warp's bytes
            const int j = it & 7;
            if (j == 0 && lane == 0)
                asm volatile("mbarrier.arrive.expect_tx.shared.b64 _, [%0], %1;" ::"r"(bar_s), "r"(32 * 8 * 32) : "memory");
            __syncwarp();
            asm volatile(
                "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], 32, [%2];" ::"r"(
                    my_s + 0u * j),
                "l"(sec), "r"(bar_s)
                : "memory");
            if (j == 7) {
                asm volatile(
                    "{\n.reg .pred P;\nW: mbarrier.try_wait.parity.shared.b64 P, [%0], %1;\n@!P bra W;\n}\n" ::"r"(bar_s),
                    "r"(phase)
                    : "memory");
                phase ^= 1;
                acc += slot[threadIdx.x * 16];
            }
        } else if (MODE == 7) {
            float v[8];
            asm volatile("ld.global.nc.v8.f32 {%0,%1,%2,%3,%4,%5,%6,%7}, [%8];"
                         : "=f"(v[0]), "=f"(v[1]), "=f"(v[2]), "=f"(v[3]), "=f"(v[4]), "=f"(v[5]), "=f"(v[6]), "=f"(v[7])
                         : "l"(sec));
            acc += v[0] + v[7];
        }
    }
    if (MODE == 3 || MODE == 4) asm volatile("cp.async.bulk.wait_group.read 0;" ::: "memory");
    if (acc == 12345.678f) sink[0] = acc;
}

template <int MODE>
double run(float* buf, uint32_t nsec, int ops, float* sink, int grid, double sectors_per_op) {
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    k<MODE><<<grid, 256>>>(buf, nsec, ops, sink);
    cudaEventRecord(e0);
    k<MODE><<<grid, 256>>>(buf, nsec, ops, sink);
    cudaEventRecord(e1);
    cudaError_t err = cudaEventSynchronize(e1);
    if (err != cudaSuccess) {
        printf("mode %d: %s\n", MODE, cudaGetErrorString(err));
        return 0;
    }
    float ms;
    cudaEventElapsedTime(&ms, e0, e1);
    // sectors touched: pairs of lanes share one
    const double threads = (double)grid * 256;
    const double sec = threads * ops * sectors_per_op;
    printf("mode %d: %.3f ms, %.3e sectors/s, %.3e thread-ops/s\n", MODE, ms, sec / (ms * 1e-3), threads * ops / (ms * 1e-3));
    cudaEventDestroy(e0);
    cudaEventDestroy(e1);
    return sec / (ms * 1e-3);
}

int main() {
    const uint32_t V = 154u * 154u * 284u;  // C2 brick image
    const uint32_t nsec = V / 8;
    float *buf, *sink;
    cudaMalloc(&buf, 4ull * V + 64);
    cudaMalloc(&sink, 64);
    cudaMemset(buf, 0, 4ull * V);
    int sms;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    for (int per : {4, 8}) {
        const int grid = sms * per;
        printf("grid %d x 256\n", grid);
        run<0>(buf, nsec, 256, sink, grid, 0.5);
        run<1>(buf, nsec, 256, sink, grid, 0.5);
        run<2>(buf, nsec, 128, sink, grid, 1.0);
        run<3>(buf, nsec, 128, sink, grid, 1.0);
        run<4>(buf, nsec, 128, sink, grid, 2.0);
        run<5>(buf, nsec, 256, sink, grid, 0.5);
        run<6>(buf, nsec, 128, sink, grid, 1.0);
        run<7>(buf, nsec, 128, sink, grid, 1.0);
    }
    return 0;
}
