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
            printf("barrier: %d blocks x %d threads: mine %.3f us, cg %.3f us  (%s)\n", blocks,
                   threads, 1e3 * ms / iters, 1e3 * ms2 / iters,
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
    return 0;
}
