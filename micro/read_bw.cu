// Pure-read HBM bandwidth on B200: the ceiling of k_hist (which only reads keys).
// nvcc -O3 -gencode arch=compute_100a,code=sm_100a -o micro/read_bw micro/read_bw.cu
// Each CTA streams a contiguous chunk with 16-byte loads (UNROLL in flight per thread)
// and folds them into one word so the loads are not dead.
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

template <int UNROLL>
__global__ void __launch_bounds__(256) rd(const uint4 *__restrict__ p, uint64_t nvec, uint32_t *out) {
    const uint64_t per = (nvec + gridDim.x - 1) / gridDim.x;
    const uint64_t b = per * blockIdx.x, e = min(nvec, b + per);
    uint32_t acc = 0;
    for (uint64_t i = b + threadIdx.x; i < e; i += 256ull * UNROLL) {
        uint4 w[UNROLL];
#pragma unroll
        for (int u = 0; u < UNROLL; ++u) {
            const uint64_t j = i + 256ull * u;
            w[u] = j < e ? __ldcs(p + j) : make_uint4(0, 0, 0, 0);
        }
#pragma unroll
        for (int u = 0; u < UNROLL; ++u) acc ^= w[u].x ^ w[u].y ^ w[u].z ^ w[u].w;
    }
    if (acc == 0x12345678u) *out = acc;
}

template <int U>
static void run(const uint4 *p, uint64_t nvec, uint32_t *o, int ctas_per_sm) {
    cudaEvent_t a, b;
    cudaEventCreate(&a);
    cudaEventCreate(&b);
    const int grid = 148 * ctas_per_sm;
    for (int i = 0; i < 3; ++i) rd<U><<<grid, 256>>>(p, nvec, o);
    float best = 1e9f;
    for (int i = 0; i < 10; ++i) {
        cudaEventRecord(a);
        rd<U><<<grid, 256>>>(p, nvec, o);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        float ms;
        cudaEventElapsedTime(&ms, a, b);
        if (ms < best) best = ms;
    }
    printf("read %llu B  unroll %2d  ctas/SM %d  best %.4f ms  %.1f GB/s\n", (unsigned long long)(nvec * 16), U,
           ctas_per_sm, best, nvec * 16 / (best * 1e6));
}

int main() {
    const uint64_t bytes = 1ull << 30;  // 2^28 u32 keys: one k_hist pass
    uint4 *p;
    uint32_t *o;
    cudaMalloc(&p, bytes);
    cudaMalloc(&o, 4);
    cudaMemset(p, 1, bytes);
    const uint64_t nvec = bytes / 16;
    for (int c : {2, 4, 8}) {
        run<4>(p, nvec, o, c);
        run<8>(p, nvec, o, c);
        run<16>(p, nvec, o, c);
    }
    return 0;
}
