// Microbenchmark (tools/, not part of libgc): sustained rate of scattered
// 64-bit global atomics with their results consumed -- the request the COUNT
// rounds issue per live entry -- over a count array the size of R-MAT s24's
// (16.8M x 8 B = 134 MB) and half of it, with Q independent atomics in flight
// per lane, every SM busy.  Reports G atomics / s (CUDA events).
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o mbr tools/microbench_atomic_rate.cu
#include <cstdio>
#include <cstdint>

__device__ __forceinline__ uint32_t mix(uint32_t x) {
    x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16;
    return x;
}

template <int Q>
__global__ void k_rate(unsigned long long *c, uint32_t n, int iters, unsigned long long *sink) {
    const uint32_t tid = blockIdx.x * blockDim.x + threadIdx.x;
    unsigned long long acc = 0;
    for (int i = 0; i < iters; ++i) {
        unsigned long long old[Q];
#pragma unroll
        for (int q = 0; q < Q; ++q) {
            const uint32_t ix = mix(tid * 0x9E3779B9u + (uint32_t)(i * Q + q) * 0x85EBCA6Bu) % n;
            asm volatile("atom.global.add.u64 %0, [%1], %2;" : "=l"(old[q]) : "l"(c + ix), "l"(1ull));
        }
#pragma unroll
        for (int q = 0; q < Q; ++q) acc += old[q];
    }
    if (acc == 0x123456789ull) *sink = acc;
}

int main() {
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    const uint32_t N = 16777216;
    unsigned long long *c, *sink;
    cudaMalloc(&c, (size_t)N * 8);
    cudaMalloc(&sink, 8);
    cudaMemset(c, 0, (size_t)N * 8);
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    for (uint32_t n : {N, N / 2, N / 8}) {
        for (int threads : {768, 1024}) {
            const int blocks = sms * (2048 / threads);
            const int iters = 64;
            k_rate<4><<<blocks, threads>>>(c, n, 4, sink);  // warm
            cudaEventRecord(e0);
            k_rate<4><<<blocks, threads>>>(c, n, iters, sink);
            cudaEventRecord(e1);
            cudaEventSynchronize(e1);
            float ms = 0;
            cudaEventElapsedTime(&ms, e0, e1);
            const double ops = (double)blocks * threads * iters * 4;
            printf("atom.add.u64 (ret), %u words (%.0f MB), %d x %d threads, 4 in flight/lane: %.2f G atomics/s\n",
                   n, n * 8.0 / 1e6, blocks, threads, ops / (ms * 1e6));
        }
    }
    return cudaGetLastError() != cudaSuccess;
}
