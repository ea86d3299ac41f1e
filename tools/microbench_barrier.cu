// Microbenchmark (tools/, not part of libgc): cost of one grid-wide barrier
// in a cooperative persistent kernel on B200, and the latency of dependent
// global loads.  nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o mb tools/microbench_barrier.cu
#include <cooperative_groups.h>
#include <cstdio>
#include <cstdint>
#include <vector>

namespace cg = cooperative_groups;

__device__ __forceinline__ bool my_barrier(unsigned long long *ctr) {
    __syncthreads();
    if (threadIdx.x == 0) {
        volatile unsigned long long *gen = ctr + 1;
        const unsigned long long g0 = *gen;
        __threadfence();
        const unsigned long long arrived = atomicAdd(ctr, 1ull) + 1;
        if (arrived == gridDim.x) {
            ctr[0] = 0;
            __threadfence();
            atomicAdd(ctr + 1, 1ull);
        } else {
            while (*gen == g0) __nanosleep(32);
        }
        __threadfence();
    }
    __syncthreads();
    return true;
}

__global__ void k_mybar(unsigned long long *ctr, int iters) {
    for (int i = 0; i < iters; ++i) my_barrier(ctr);
}

// the kernel's barrier: monotone counter, fence + relaxed atomic, acquire
// spin, trailing fence
__device__ __forceinline__ unsigned long long ld_acq(const unsigned long long *p) {
    unsigned long long v;
    asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ unsigned long long atom_add_rel(unsigned long long *p, unsigned long long x) {
    unsigned long long v;
    asm volatile("atom.add.release.gpu.global.u64 %0, [%1], %2;" : "=l"(v) : "l"(p), "l"(x) : "memory");
    return v;
}
__global__ void k_monobar(unsigned long long *ctr, int iters) {
    for (int i = 0; i < iters; ++i) {
        __syncthreads();
        if (threadIdx.x == 0) {
            __threadfence();
            const unsigned long long old = atomicAdd(ctr, 1ull);
            const unsigned long long target = (old / gridDim.x + 1) * gridDim.x;
            while (ld_acq(ctr) < target) {
            }
            __threadfence();
        }
        __syncthreads();
    }
}
// release-atomic arrival, acquire spin, no explicit fences
__global__ void k_relbar(unsigned long long *ctr, int iters) {
    for (int i = 0; i < iters; ++i) {
        __syncthreads();
        if (threadIdx.x == 0) {
            const unsigned long long old = atom_add_rel(ctr, 1ull);
            const unsigned long long target = (old / gridDim.x + 1) * gridDim.x;
            while (ld_acq(ctr) < target) {
            }
        }
        __syncthreads();
    }
}

__global__ void k_cgbar(int iters) {
    cg::grid_group g = cg::this_grid();
    for (int i = 0; i < iters; ++i) g.sync();
}

// pointer chase: each step loads the next index (dependent loads)
__global__ void k_chase(const uint32_t *next, int steps, uint32_t *out, int start) {
    uint32_t p = start;
    for (int i = 0; i < steps; ++i) p = next[p];
    *out = p;
}

// every warp chases its own random chain through a big array (loaded GPU)
__global__ void k_chase_many(const uint32_t *next, size_t n, int steps, uint32_t *out) {
    const unsigned lane = threadIdx.x & 31;
    uint32_t p = (uint32_t)(((blockIdx.x * blockDim.x + threadIdx.x) >> 5) * 2654435761u % n);
    if (lane == 0)
        for (int i = 0; i < steps; ++i) p = next[p];
    if (lane == 0 && p == 0xFFFFFFFFu) *out = p;
}

// cost of __threadfence with outstanding stores
__global__ void k_fence(uint32_t *buf, int iters, unsigned long long *cyc) {
    unsigned long long t0 = clock64();
    for (int i = 0; i < iters; ++i) {
        buf[(threadIdx.x + i * 977) & 0xFFFFF] = i;
        __threadfence();
    }
    if (threadIdx.x == 0) cyc[blockIdx.x] = clock64() - t0;
}

int main() {
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    unsigned long long *ctr;
    cudaMalloc(&ctr, 64);
    cudaEvent_t a, b;
    cudaEventCreate(&a);
    cudaEventCreate(&b);
    for (int threads : {256, 512, 1024}) {
        int per = 0;
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per, k_mybar, threads, 0);
        for (int bps : {1, per}) {
            int blocks = sms * bps;
            int iters = 2000;
            cudaMemset(ctr, 0, 64);
            void *args[] = {&ctr, &iters};
            cudaLaunchCooperativeKernel((void *)k_mybar, blocks, threads, args, 0, 0);
            cudaEventRecord(a);
            cudaLaunchCooperativeKernel((void *)k_mybar, blocks, threads, args, 0, 0);
            cudaEventRecord(b);
            cudaEventSynchronize(b);
            float ms;
            cudaEventElapsedTime(&ms, a, b);
            void *args2[] = {&iters};
            cudaLaunchCooperativeKernel((void *)k_cgbar, blocks, threads, args2, 0, 0);
            cudaEventRecord(a);
            cudaLaunchCooperativeKernel((void *)k_cgbar, blocks, threads, args2, 0, 0);
            cudaEventRecord(b);
            cudaEventSynchronize(b);
            float ms2;
            cudaEventElapsedTime(&ms2, a, b);
            float ms3, ms4;
            cudaMemset(ctr, 0, 64);
            cudaLaunchCooperativeKernel((void *)k_monobar, blocks, threads, args, 0, 0);
            cudaEventRecord(a);
            cudaLaunchCooperativeKernel((void *)k_monobar, blocks, threads, args, 0, 0);
            cudaEventRecord(b);
            cudaEventSynchronize(b);
            cudaEventElapsedTime(&ms3, a, b);
            cudaMemset(ctr, 0, 64);
            cudaLaunchCooperativeKernel((void *)k_relbar, blocks, threads, args, 0, 0);
            cudaEventRecord(a);
            cudaLaunchCooperativeKernel((void *)k_relbar, blocks, threads, args, 0, 0);
            cudaEventRecord(b);
            cudaEventSynchronize(b);
            cudaEventElapsedTime(&ms4, a, b);
            printf("barrier: %d blocks x %d threads: gen %.3f us, mono+fences %.3f us, "
                   "release/acquire %.3f us, cg %.3f us  (%s)\n", blocks, threads,
                   1e3 * ms / iters, 1e3 * ms3 / iters, 1e3 * ms4 / iters, 1e3 * ms2 / iters,
                   cudaGetErrorString(cudaGetLastError()));
        }
    }
    // dependent loads: random permutation cycle in a buffer of `sz` words
    for (size_t sz : {(size_t)1 << 16, (size_t)1 << 22, (size_t)1 << 26}) {
        std::vector<uint32_t> h(sz);
        for (size_t i = 0; i < sz; ++i) h[i] = (uint32_t)i;
        uint64_t x = 88172645463325252ull;
        for (size_t i = sz - 1; i > 0; --i) {
            x ^= x << 13; x ^= x >> 7; x ^= x << 17;
            size_t j = x % (i + 1);
            std::swap(h[i], h[j]);
        }
        std::vector<uint32_t> nxt(sz);
        for (size_t i = 0; i < sz; ++i) nxt[h[i]] = h[(i + 1) % sz];
        uint32_t *d, *o;
        cudaMalloc(&d, sz * 4);
        cudaMalloc(&o, 4);
        cudaMemcpy(d, nxt.data(), sz * 4, cudaMemcpyHostToDevice);
        int steps = 20000;
        k_chase<<<1, 1>>>(d, 1000, o, 0);
        cudaEventRecord(a);
        k_chase<<<1, 1>>>(d, steps, o, 0);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        float ms;
        cudaEventElapsedTime(&ms, a, b);
        printf("dependent load chain, %zu MB working set: %.1f ns per load\n", sz * 4 >> 20,
               1e6 * ms / steps);
        cudaFree(d);
        cudaFree(o);
    }
    {
        size_t n = (size_t)1 << 29;  // 2 GiB of uint32
        uint32_t *d, *o;
        cudaMalloc(&d, n * 4);
        cudaMalloc(&o, 4);
        // next[i] = hash(i) mod n: a random functional graph (good enough)
        std::vector<uint32_t> h(1 << 20);
        for (size_t c = 0; c < n; c += h.size()) {
            for (size_t i = 0; i < h.size(); ++i) {
                uint64_t x = (c + i) * 0x9E3779B97F4A7C15ull;
                x ^= x >> 29; x *= 0xBF58476D1CE4E5B9ull; x ^= x >> 32;
                h[i] = (uint32_t)(x % n);
            }
            cudaMemcpy(d + c, h.data(), h.size() * 4, cudaMemcpyHostToDevice);
        }
        int sms = 0;
        cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
        for (int warps_per_sm : {1, 8, 32}) {
            int steps = 2000;
            k_chase_many<<<sms, 32 * warps_per_sm>>>(d, n, 100, o);
            cudaEventRecord(a);
            k_chase_many<<<sms, 32 * warps_per_sm>>>(d, n, steps, o);
            cudaEventRecord(b);
            cudaEventSynchronize(b);
            float ms;
            cudaEventElapsedTime(&ms, a, b);
            printf("loaded chase, 2 GiB, %d warps/SM (%d warps): %.1f ns per dependent load\n",
                   warps_per_sm, warps_per_sm * sms, 1e6 * ms / steps);
        }
        unsigned long long *cyc;
        cudaMalloc(&cyc, sizeof(unsigned long long) * sms);
        k_fence<<<sms, 32>>>(d, 1000, cyc);
        cudaEventRecord(a);
        k_fence<<<sms, 32>>>(d, 1000, cyc);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        float ms;
        cudaEventElapsedTime(&ms, a, b);
        printf("store + __threadfence: %.1f ns per iteration (1 warp/SM)\n", 1e6 * ms / 1000);
        cudaFree(d);
    }
    return 0;
}
