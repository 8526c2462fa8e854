// Debug harness: prints lor_setup / slab_pieces intermediates for one event (tools only).
#include <cstdio>
#include "lmosem_kernels.cuh"
using namespace lmk;
__global__ void k(const float* ev, GridGeom g) {
    Lor L;
    bool ok = lor_setup(ev, g, L);
    printf("ok %d i0 %d ns %d code %d fin %.9g fout %.9g lunit %.9g ab %.9g ac %.9g\n", ok, L.i0, L.ns, L.code,
           L.fin, L.fout, L.lunit, L.ab, L.ac);
    printf("wb0 %lld sb %lld wc0 %lld sc %lld\n", L.wb0, L.sb, L.wc0, L.sc);
    Walk W = make_walk(L, g);
    Step S = make_step(L, W, 0);
    Pieces P = slab_pieces(L, W, 0, S.wb, S.wc, S.Ja);
    printf("l0 %.9g l1 %.9g l2 %.9g j %d %d %d\n", P.l0, P.l1, P.l2, P.j0, P.j1, P.j2);
}
int main() {
    float h[6] = {-4.885164f, -18.939774f, -5.6115713f, -12.046729f, 9.170044f, -23.146145f};
    int dims[3] = {33, 5, 64};
    float vox[3] = {0.6f, 2.0f, 0.45f};
    GridGeom g{};
    for (int q = 0; q < 3; ++q) {
        g.n[q] = dims[q];
        g.lo[q] = -0.5 * dims[q] * (double)vox[q];
        g.inv_v[q] = 1.0 / (double)vox[q];
        g.clo[q] = 0;
        g.chi[q] = dims[q];
        g.P[q] = (dims[q] + 5) & ~1;
    }
    int64_t M[3] = {8, 8LL * g.P[0] / 2, 8LL * g.P[0] / 2 * g.P[1] / 2}, m[3] = {1, 2, 4};
    for (int q = 0; q < 3; ++q) { g.A[q] = (int)(M[q] / 2); g.B[q] = (int)(m[q] - M[q] / 2); }
    float* d;
    cudaMalloc(&d, 24);
    cudaMemcpy(d, h, 24, cudaMemcpyHostToDevice);
    k<<<1, 1>>>(d, g);
    cudaDeviceSynchronize();
    return 0;
}
