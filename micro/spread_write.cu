// Is the first scatter pass slow because its 256 write streams are 4 MB apart?
// Write-only model of a scatter's write-out: 2^28 4-byte elements, NS = 256 streams,
// "tile" t writes run [t*R, (t+1)*R) of every stream (R = 28 records, the c2 tile
// 7168 / 256), tiles claimed in order by a persistent grid (2 CTAs/SM x 256 threads,
// one warp per run).  Layouts:
//   spread   stream s at s * 4 MB (pass 1: one bucket -> 256 sub-buckets)
//   spreadp  stream s at s * (4 MB + 4 KB + 64 B) (no power-of-two stride)
//   local    streams grouped: bucket b = 4 MB region, 256 sub-streams 16 KB apart,
//            tiles walk one bucket at a time (pass 2)
// nvcc -O3 -gencode arch=compute_100a,code=sm_100a -o micro/spread_write micro/spread_write.cu
#include <cstdio>
#include <cstdint>
#include <cuda.h>
#include <cuda_runtime.h>

constexpr int NS = 256, R = 28;

__global__ void __launch_bounds__(256) wr(uint32_t *out, uint64_t n, int mode, uint64_t stride, unsigned *claim) {
    const uint64_t per_stream = n / NS;                 // elements per stream (spread modes)
    const uint64_t tiles = n / (uint64_t(NS) * R);      // tiles
    __shared__ unsigned t_s;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    for (;;) {
        if (threadIdx.x == 0) t_s = atomicAdd(claim, 1u);
        __syncthreads();
        const uint64_t t = t_s;
        __syncthreads();
        if (t >= tiles) break;
        // per-tile bucket / run of the pass-2 layouts (hoisted: 64-bit divisions per store would
        // make the model compute-bound)
        uint64_t b2 = 0, k2 = 0;
        bool skip2 = false;
        if (mode == 100) {
            const uint64_t tpb = (uint64_t(1) << 20) / (uint64_t(NS) * R) + 1;
            b2 = t / tpb;
            k2 = t % tpb;
        } else if (mode >= 2) {
            // buckets of 2^20 records (4 MB), 256 sub-streams of 2^12 records (16 KB) each;
            // G = mode - 1 buckets in flight at once (consecutive tiles alternate between
            // them): about 2 G pages written at a time
            const uint64_t G = mode - 1;
            const uint64_t tpb = ((uint64_t(1) << 12) + R - 1) / R;  // tiles per bucket
            const uint64_t grp = t / (G * tpb), j = t % (G * tpb);
            b2 = grp * G + j % G;
            k2 = j / G;
            skip2 = b2 >= NS || (k2 + 1) * R > (uint64_t(1) << 12);
        }
        for (int s = warp; s < NS; s += 8) {
            uint64_t base;
            if (mode == 100) {  // the first version of the pass-2 model (tile 146 of a bucket overlaps)
                base = b2 * (uint64_t(1) << 20) + s * (uint64_t(1) << 12) + k2 * R;
                if (base + R > n) continue;
            } else if (mode >= 2) {
                if (skip2) continue;
                base = b2 * (uint64_t(1) << 20) + s * (uint64_t(1) << 12) + k2 * R;
            } else {
                base = s * stride + t * R;
                if (t * R + R > per_stream) continue;
            }
            if (lane < R) out[base + lane] = static_cast<uint32_t>(t + lane);
        }
    }
}

// device memory through the VMM API: physical chunks of `gran` bytes mapped at an address
// aligned to `align` (does the GMMU use larger TLB entries for larger aligned mappings?)
static uint32_t *vmm_alloc(size_t bytes, size_t gran, size_t align) {
    CUmemAllocationProp prop = {};
    prop.type = CU_MEM_ALLOCATION_TYPE_PINNED;
    prop.location.type = CU_MEM_LOCATION_TYPE_DEVICE;
    prop.location.id = 0;
    bytes = (bytes + gran - 1) / gran * gran;
    CUdeviceptr va;
    if (cuMemAddressReserve(&va, bytes, align, 0, 0) != CUDA_SUCCESS) return nullptr;
    CUmemGenericAllocationHandle h;
    if (cuMemCreate(&h, bytes, &prop, 0) != CUDA_SUCCESS) return nullptr;
    if (cuMemMap(va, bytes, 0, h, 0) != CUDA_SUCCESS) return nullptr;
    CUmemAccessDesc ad = {};
    ad.location = prop.location;
    ad.flags = CU_MEM_ACCESS_FLAGS_PROT_READWRITE;
    if (cuMemSetAccess(va, bytes, &ad, 1) != CUDA_SUCCESS) return nullptr;
    return reinterpret_cast<uint32_t *>(va);
}

static void sweep(const char *tag, uint32_t *out, uint64_t n, unsigned *claim) {
    const uint64_t strides[] = {n / NS, n / NS + 1024 + 16};
    const int groups[] = {1, 4, 16, 64, 128};
    for (int m = 0; m < 8; ++m) {
        const int mode = m < 2 ? 1 : m == 7 ? 100 : 1 + groups[m - 2];
        float best = 1e9f;
        for (int i = 0; i < 6; ++i) {
            cudaMemset(claim, 0, 4);
            cudaEvent_t a, b;
            cudaEventCreate(&a);
            cudaEventCreate(&b);
            cudaEventRecord(a);
            wr<<<296, 256>>>(out, n, mode, m < 2 ? strides[m] : 0, claim);
            cudaEventRecord(b);
            cudaEventSynchronize(b);
            float ms;
            cudaEventElapsedTime(&ms, a, b);
            if (i > 0 && ms < best) best = ms;
        }
        if (m < 2)
            printf("%s pass-1 layout, stride %llu B        best %.4f ms  %.1f GB/s written\n", tag,
                   (unsigned long long)(strides[m] * 4), best, n * 4 / (best * 1e6));
        else if (m == 7)
            printf("%s pass-2 layout, first model             best %.4f ms  %.1f GB/s written\n", tag, best,
                   n * 4 / (best * 1e6));
        else
            printf("%s pass-2 layout, %3d buckets in flight best %.4f ms  %.1f GB/s written\n", tag, groups[m - 2],
                   best, n * 4 / (best * 1e6));
    }
}

int main() {
    const uint64_t n = 1ull << 28;
    cudaFree(0);
    unsigned *claim;
    cudaMalloc(&claim, 4);
    CUmemAllocationProp prop = {};
    prop.type = CU_MEM_ALLOCATION_TYPE_PINNED;
    prop.location.type = CU_MEM_LOCATION_TYPE_DEVICE;
    prop.location.id = 0;
    size_t gmin = 0, grec = 0;
    cuMemGetAllocationGranularity(&gmin, &prop, CU_MEM_ALLOC_GRANULARITY_MINIMUM);
    cuMemGetAllocationGranularity(&grec, &prop, CU_MEM_ALLOC_GRANULARITY_RECOMMENDED);
    printf("VMM granularity: minimum %zu, recommended %zu\n", gmin, grec);
    uint32_t *out;
    cudaMalloc(&out, n * 4 + (64ull << 20));
    sweep("cudaMalloc   ", out, n, claim);
    for (size_t align : {size_t(2) << 20, size_t(512) << 20, size_t(1) << 30}) {
        uint32_t *o = vmm_alloc(n * 4 + (64ull << 20), gmin, align);
        if (!o) { printf("vmm alloc (align %zu) failed\n", align); continue; }
        char tag[64];
        snprintf(tag, sizeof tag, "vmm %4zu MB al", align >> 20);
        sweep(tag, o, n, claim);
    }
    cudaError_t e = cudaGetLastError();
    if (e != cudaSuccess) printf("error %s\n", cudaGetErrorString(e));
    return 0;
}
