// Microbenchmarks (not part of the library): histogram counting strategies and stable
// in-tile ranking strategies on B200, 2^28 uint32 keys resident in HBM.
#include <cstdio>
#include <cstdint>
#include <cstdlib>
#include <vector>
#include <cuda_runtime.h>

#define CK(x) do { cudaError_t e = (x); if (e != cudaSuccess) { printf("CUDA %s at %d\n", cudaGetErrorString(e), __LINE__); exit(1);} } while (0)

__device__ __forceinline__ uint32_t lanemask_lt() { uint32_t r; asm("mov.u32 %0, %%lanemask_lt;" : "=r"(r)); return r; }

// ---------------------------------------------------------------- read-only reference
__global__ void k_read(const uint4* __restrict__ in, size_t nvec, uint32_t* out) {
  uint32_t acc = 0;
  for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < nvec; i += (size_t)gridDim.x * blockDim.x) {
    uint4 v = __ldg(in + i); acc ^= v.x ^ v.y ^ v.z ^ v.w;
  }
  if (acc == 0x12345678) out[0] = acc;
}
__global__ void k_copy(const uint4* __restrict__ in, uint4* __restrict__ out, size_t nvec) {
  for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < nvec; i += (size_t)gridDim.x * blockDim.x) out[i] = __ldg(in + i);
}

// ---------------------------------------------------------------- histogram variants
template <int MODE>
__global__ void __launch_bounds__(512) k_hist(const uint4* __restrict__ in, size_t nvec, uint32_t* out, int shift) {
  __shared__ uint32_t h[16][256];
  const int w = threadIdx.x >> 5;
  for (int i = threadIdx.x; i < 16 * 256; i += blockDim.x) (&h[0][0])[i] = 0;
  __syncthreads();
  uint32_t* my = MODE == 3 ? h[0] : h[w];
  const size_t stride = (size_t)gridDim.x * blockDim.x;
  size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x;
  // uniform trip count per warp so match has all lanes
  const size_t iters = (nvec + stride - 1) / stride;
  for (size_t it = 0; it < iters; it += 4) {
    uint4 v[4]; bool ok[4];
#pragma unroll
    for (int u = 0; u < 4; ++u) { size_t j = i + (it + u) * stride; ok[u] = (it + u < iters) && j < nvec; if (ok[u]) v[u] = __ldg(in + j); }
#pragma unroll
    for (int u = 0; u < 4; ++u) {
      uint32_t d[4] = {(v[u].x >> shift) & 255, (v[u].y >> shift) & 255, (v[u].z >> shift) & 255, (v[u].w >> shift) & 255};
      if (MODE == 0 || MODE == 3) {  // plain atomics
        if (ok[u]) {
#pragma unroll
          for (int k = 0; k < 4; ++k) atomicAdd(&my[d[k]], 1u);
        }
      } else if (MODE == 1) {  // warp match aggregation, predicated
#pragma unroll
        for (int k = 0; k < 4; ++k) {
          uint32_t dd = ok[u] ? d[k] : 256u;
          uint32_t m = __match_any_sync(0xffffffffu, dd);
          bool lead = ((m & lanemask_lt()) == 0) && dd < 256;
          if (lead) atomicAdd(&my[dd], (uint32_t)__popc(m));
        }
      } else if (MODE == 2) {  // in-thread combine of equal neighbours
        if (ok[u]) {
          if (d[0] == d[1] && d[1] == d[2] && d[2] == d[3]) atomicAdd(&my[d[0]], 4u);
          else {
#pragma unroll
            for (int k = 0; k < 4; ++k) atomicAdd(&my[d[k]], 1u);
          }
        }
      } else if (MODE == 4) {  // packed: 2 digits per atomic via 16-bit halves (bin pairs)
        if (ok[u]) {
#pragma unroll
          for (int k = 0; k < 4; ++k) atomicAdd(&my[d[k] >> 1], 1u << ((d[k] & 1) * 16));
        }
      }
    }
  }
  __syncthreads();
  for (int b = threadIdx.x; b < 256; b += blockDim.x) {
    uint32_t s = 0;
    for (int q = 0; q < 16; ++q) s += h[q][b];
    atomicAdd(&out[b], s);
  }
}

// ---------------------------------------------------------------- in-tile stable rank variants
// Each CTA: THREADS x KPT keys (warp-striped), rank by digit, write the locally partitioned
// tile back contiguously (no global scatter) -> measures load + rank + staged store.
template <int THREADS, int KPT, int MODE>
__global__ void __launch_bounds__(THREADS) k_rank(const uint32_t* __restrict__ in, uint32_t* __restrict__ out, size_t n, int shift) {
  constexpr int W = THREADS / 32, KPB = THREADS * KPT, NB = 257;
  extern __shared__ uint32_t sm[];
  uint32_t* wcnt = sm;              // W * NB
  uint32_t* tot = sm + W * NB;      // NB (+pad)
  uint32_t* sk = tot + 288;         // KPB
  const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
  const uint32_t ltm = lanemask_lt();
  const size_t ntiles = n / KPB;
  for (size_t t = blockIdx.x; t < ntiles; t += gridDim.x) {
    const uint32_t* src = in + t * KPB;
    uint32_t key[KPT], rk[KPT];
#pragma unroll
    for (int c = 0; c < KPT; ++c) key[c] = src[warp * 32 * KPT + c * 32 + lane];
    for (int i = tid; i < W * NB; i += THREADS) wcnt[i] = 0;
    if (t == blockIdx.x) for (int i = tid; i < W * 512; i += THREADS) sm[W * NB + 288 + KPB + i] = 0;
    __syncthreads();
    uint32_t* my = wcnt + warp * NB;
    if (MODE == 0) {  // match walk
#pragma unroll
      for (int c = 0; c < KPT; ++c) {
        uint32_t d = (key[c] >> shift) & 255;
        uint32_t m = __match_any_sync(0xffffffffu, d);
        uint32_t below = m & ltm;
        uint32_t pre = my[d];
        __syncwarp();
        if (below == 0) my[d] = pre + __popc(m);
        __syncwarp();
        rk[c] = ((pre + __popc(below)) << 9) | d;
      }
    } else if (MODE == 1) {  // bit-sliced ballots
#pragma unroll
      for (int c = 0; c < KPT; ++c) {
        uint32_t d = (key[c] >> shift) & 255;
        uint32_t m = 0xffffffffu;
#pragma unroll
        for (int b = 0; b < 8; ++b) {
          uint32_t bal = __ballot_sync(0xffffffffu, (d >> b) & 1);
          m &= ((d >> b) & 1) ? bal : ~bal;
        }
        uint32_t below = m & ltm;
        uint32_t pre = my[d];
        __syncwarp();
        if (below == 0) my[d] = pre + __popc(m);
        __syncwarp();
        rk[c] = ((pre + __popc(below)) << 9) | d;
      }
    } else if (MODE == 3) {  // peer mask via smem atomicOr, running count via leader atomicAdd + shfl
      uint32_t* pm = sm + W * NB + 288 + KPB + warp * 256;
#pragma unroll
      for (int c = 0; c < KPT; ++c) {
        uint32_t d = (key[c] >> shift) & 255;
        atomicOr(&pm[d], 1u << lane);
        __syncwarp();
        uint32_t m = pm[d];
        __syncwarp();
        pm[d] = 0;
        int leader = __ffs(m) - 1;
        uint32_t pre = 0;
        if (lane == leader) pre = atomicAdd(&my[d], (uint32_t)__popc(m));
        pre = __shfl_sync(0xffffffffu, pre, leader);
        rk[c] = ((pre + __popc(m & ltm)) << 9) | d;
      }
    } else if (MODE == 4) {  // peer mask via smem atomicOr, running count via LDS/STS
      uint32_t* pm = sm + W * NB + 288 + KPB + warp * 256;
#pragma unroll
      for (int c = 0; c < KPT; ++c) {
        uint32_t d = (key[c] >> shift) & 255;
        atomicOr(&pm[d], 1u << lane);
        __syncwarp();
        uint32_t m = pm[d];
        uint32_t pre = my[d];
        __syncwarp();
        uint32_t below = m & ltm;
        if (below == 0) { my[d] = pre + __popc(m); pm[d] = 0; }
        __syncwarp();
        rk[c] = ((pre + __popc(below)) << 9) | d;
      }
    } else if (MODE == 5) {  // peer mask via NON-returning atomicAdd(1<<lane) (sum == or), count LDS/STS
      uint32_t* pm = sm + W * NB + 288 + KPB + warp * 256;
#pragma unroll
      for (int c = 0; c < KPT; ++c) {
        uint32_t d = (key[c] >> shift) & 255;
        atomicAdd(&pm[d], 1u << lane);
        __syncwarp();
        uint32_t m = pm[d];
        uint32_t pre = my[d];
        __syncwarp();
        uint32_t below = m & ltm;
        if (below == 0) { my[d] = pre + __popc(m); pm[d] = 0; }
        __syncwarp();
        rk[c] = ((pre + __popc(below)) << 9) | d;
      }
    } else if (MODE == 6) {  // packed 64-bit {count:32 | mask:32}, non-returning atomicAdd
      unsigned long long* pk = reinterpret_cast<unsigned long long*>(sm + W * NB + 288 + KPB) + warp * 256;
#pragma unroll
      for (int c = 0; c < KPT; ++c) {
        uint32_t d = (key[c] >> shift) & 255;
        atomicAdd(&pk[d], 1ull << lane);
        __syncwarp();
        unsigned long long v = pk[d];
        __syncwarp();
        uint32_t m = (uint32_t)v, pre = (uint32_t)(v >> 32);
        uint32_t below = m & ltm;
        if (below == 0) pk[d] = (unsigned long long)(pre + __popc(m)) << 32;
        __syncwarp();
        rk[c] = ((pre + __popc(below)) << 9) | d;
      }
      __syncwarp();
      for (int d = lane; d < 256; d += 32) { my[d] = (uint32_t)(pk[d] >> 32); pk[d] = 0; }
    } else if (MODE == 7) {  // count via non-returning atomics, match only among lanes with duplicates
#pragma unroll
      for (int c = 0; c < KPT; ++c) {
        uint32_t d = (key[c] >> shift) & 255;
        uint32_t pre = my[d];
        __syncwarp();
        atomicAdd(&my[d], 1u);
        __syncwarp();
        uint32_t k = my[d] - pre;
        uint32_t r = 0;
        uint32_t dup = __ballot_sync(0xffffffffu, k > 1);
        if (k > 1) {
          uint32_t m = __match_any_sync(dup, d);
          r = __popc(m & ltm);
        }
        rk[c] = ((pre + r) << 9) | d;
      }
    } else if (MODE == 8) {  // bit-sliced ballots, leader returning atomicAdd + shfl
#pragma unroll
      for (int c = 0; c < KPT; ++c) {
        uint32_t d = (key[c] >> shift) & 255;
        uint32_t m = 0xffffffffu;
#pragma unroll
        for (int b = 0; b < 8; ++b) {
          uint32_t bal = __ballot_sync(0xffffffffu, (d >> b) & 1);
          m &= ((d >> b) & 1) ? bal : ~bal;
        }
        const int leader = __ffs(m) - 1;
        uint32_t pre = 0;
        if (lane == leader) pre = atomicAdd(&my[d], (uint32_t)__popc(m));
        pre = __shfl_sync(0xffffffffu, pre, leader);
        rk[c] = ((pre + __popc(m & ltm)) << 9) | d;
      }
    } else if (MODE == 9) {  // ballots with xor-trick mask, leader returning atomicAdd + shfl
#pragma unroll
      for (int c = 0; c < KPT; ++c) {
        uint32_t d = (key[c] >> shift) & 255;
        uint32_t m = 0xffffffffu;
#pragma unroll
        for (int b = 0; b < 8; ++b) {
          uint32_t bal = __ballot_sync(0xffffffffu, (d >> b) & 1);
          m &= bal ^ (((d >> b) & 1) - 1u);
        }
        const int leader = __ffs(m) - 1;
        uint32_t pre = 0;
        if (lane == leader) pre = atomicAdd(&my[d], (uint32_t)__popc(m));
        pre = __shfl_sync(0xffffffffu, pre, leader);
        rk[c] = ((pre + __popc(m & ltm)) << 9) | d;
      }
    } else {  // MODE 2: unstable reference: atomicAdd returning old (NOT stable; cost reference only)
#pragma unroll
      for (int c = 0; c < KPT; ++c) {
        uint32_t d = (key[c] >> shift) & 255;
        rk[c] = (atomicAdd(&my[d], 1u) << 9) | d;
      }
    }
    __syncthreads();
    for (int d = tid; d < NB; d += THREADS) {
      uint32_t run = 0;
#pragma unroll
      for (int w = 0; w < W; ++w) { uint32_t v = wcnt[w * NB + d]; wcnt[w * NB + d] = run; run += v; }
      tot[d] = run;
    }
    __syncthreads();
    if (tid < 32) {
      uint32_t v[9], s = 0;
#pragma unroll
      for (int i = 0; i < 9; ++i) { int idx = lane * 9 + i; v[i] = idx < NB ? tot[idx] : 0; s += v[i]; }
      uint32_t incl = s;
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) { uint32_t y = __shfl_up_sync(0xffffffffu, incl, o); if (lane >= o) incl += y; }
      uint32_t run = incl - s;
#pragma unroll
      for (int i = 0; i < 9; ++i) { int idx = lane * 9 + i; if (idx < NB) tot[idx] = run; run += v[i]; }
    }
    __syncthreads();
    for (int d = tid; d < NB; d += THREADS) { uint32_t ls = tot[d];
#pragma unroll
      for (int w = 0; w < W; ++w) wcnt[w * NB + d] += ls; }
    __syncthreads();
#pragma unroll
    for (int c = 0; c < KPT; ++c) { uint32_t d = rk[c] & 511; sk[my[d] + (rk[c] >> 9)] = key[c]; }
    __syncthreads();
    uint32_t* dst = out + t * KPB;
#pragma unroll
    for (int c = 0; c < KPT; ++c) dst[c * THREADS + tid] = sk[c * THREADS + tid];
    __syncthreads();
  }
}

// ---------------------------------------------------------------- driver
__global__ void k_gen(uint32_t* k, size_t n, int m) {
  for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n; i += (size_t)gridDim.x * blockDim.x) {
    uint32_t acc = 0xffffffffu;
    if (m == 0) acc = 0;
    for (int j = 0; j < m; ++j) { uint64_t z = i * 0x9E3779B97F4A7C15ull + j * 0xD1B54A32D192ED03ull + 0x1234567ull;
      z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull; z = (z ^ (z >> 27)) * 0x94D049BB133111EBull; z ^= z >> 31; acc &= (uint32_t)z; }
    k[i] = acc;
  }
}

__global__ void k_cmp(const uint32_t* a, const uint32_t* b, size_t n, unsigned long long* bad) {
  unsigned long long c = 0;
  for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n; i += (size_t)gridDim.x * blockDim.x) c += a[i] != b[i];
  if (c) atomicAdd(bad, c);
}

template <typename F>
float timeit(F f, int reps = 5) {
  cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
  f(); f(); CK(cudaDeviceSynchronize());
  cudaEventRecord(a);
  for (int r = 0; r < reps; ++r) f();
  cudaEventRecord(b); CK(cudaEventSynchronize(b));
  float ms; cudaEventElapsedTime(&ms, a, b); return ms / reps;
}

int main() {
  const size_t n = 1ull << 28;
  uint32_t *keys, *out, *hist;
  CK(cudaMalloc(&keys, n * 4)); CK(cudaMalloc(&out, n * 4)); CK(cudaMalloc(&hist, 1024 * 4));
  int sms; cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  const size_t nvec = n / 4;
  const char* dname[] = {"const", "uniform", "and2", "and3", "and4"};
  int dm[] = {0, 1, 2, 3, 4};
  float ms = timeit([&] { k_read<<<sms * 4, 512>>>((const uint4*)keys, nvec, hist); });
  printf("read-only 1 GiB: %.3f ms  %.0f GB/s\n", ms, n * 4 / ms / 1e6);
  ms = timeit([&] { k_copy<<<sms * 4, 512>>>((const uint4*)keys, (uint4*)out, nvec); });
  printf("copy 1 GiB: %.3f ms  %.0f GB/s (r+w)\n", ms, 2 * n * 4 / ms / 1e6);
  for (int di = 0; di < 5; ++di) {
    k_gen<<<sms * 8, 256>>>(keys, n, dm[di]); CK(cudaDeviceSynchronize());
    for (int occ = 2; occ <= 0; occ += 2) {
      float t0 = timeit([&] { k_hist<0><<<sms * occ, 512>>>((const uint4*)keys, nvec, hist, 24); });
      float t1 = timeit([&] { k_hist<1><<<sms * occ, 512>>>((const uint4*)keys, nvec, hist, 24); });
      float t2 = timeit([&] { k_hist<2><<<sms * occ, 512>>>((const uint4*)keys, nvec, hist, 24); });
      float t3 = timeit([&] { k_hist<3><<<sms * occ, 512>>>((const uint4*)keys, nvec, hist, 24); });
      float t4 = timeit([&] { k_hist<4><<<sms * occ, 512>>>((const uint4*)keys, nvec, hist, 24); });
      printf("hist %-7s occ%d: warp-atomics %.3f ms (%.0f GB/s) | match %.3f (%.0f) | combine4 %.3f (%.0f) | block-atomics %.3f (%.0f) | packed16 %.3f (%.0f)\n",
             dname[di], occ, t0, n * 4 / t0 / 1e6, t1, n * 4 / t1 / 1e6, t2, n * 4 / t2 / 1e6, t3, n * 4 / t3 / 1e6, t4, n * 4 / t4 / 1e6);
    }
    {
      auto run = [&](auto kern, int threads, int kpt, const char* name) {
        size_t smem = (threads / 32 * 257 + 288 + threads * kpt + threads / 32 * 512) * 4;
        cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        int per = 0; cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per, kern, threads, smem);
        float t = timeit([&] { kern<<<sms * per, threads, smem>>>(keys, out, n, 24); });
        printf("rank %-7s %-22s occ%d: %.3f ms  %.0f GB/s (r+w keys)\n", dname[di], name, per, t, 2.0 * n * 4 / t / 1e6);
      };
      {
        uint32_t* ref; unsigned long long* bad;
        CK(cudaMalloc(&ref, n * 4)); CK(cudaMalloc(&bad, 8));
        for (int shift : {0, 8, 16, 24}) {
          auto go = [&](auto kern, uint32_t* o) {
            size_t smem = (256 / 32 * 257 + 288 + 256 * 16 + 256 / 32 * 512) * 4;
            cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
            kern<<<sms * 3, 256, smem>>>(keys, o, n, shift);
          };
          go(k_rank<256, 16, 7>, ref);
          go(k_rank<256, 16, 2>, out);
          cudaMemset(bad, 0, 8);
          k_cmp<<<sms * 4, 512>>>(ref, out, n, bad);
          unsigned long long hb = 0; CK(cudaMemcpy(&hb, bad, 8, cudaMemcpyDeviceToHost));
          printf("order check %-7s shift %2d: returning-atomic rank differs from stable rank at %llu of %zu\n", dname[di], shift, hb, n);
        }
        cudaFree(ref); cudaFree(bad);
      }
      continue;
      run(k_rank<256, 16, 0>, 256, 16, "match 256x16");
      run(k_rank<256, 16, 2>, 256, 16, "atomic(unstable) 256x16");
      run(k_rank<256, 16, 7>, 256, 16, "cnt+dupmatch 256x16");
      run(k_rank<256, 16, 1>, 256, 16, "ballot+lds 256x16");
      run(k_rank<256, 16, 8>, 256, 16, "ballot+ratom 256x16");
      run(k_rank<256, 16, 9>, 256, 16, "ballotx+ratom 256x16");
      run(k_rank<256, 8, 9>, 256, 8, "ballotx+ratom 256x8");
      run(k_rank<512, 8, 9>, 512, 8, "ballotx+ratom 512x8");
    }
  }
  return 0;
}
