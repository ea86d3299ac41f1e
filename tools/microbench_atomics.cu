// Microbenchmark (tools/, not part of libgc): latency of a burst of scattered
// global atomics / loads issued by every warp of a persistent grid at once --
// the access pattern of one COUNT-mode round (each warp: 8 independent random
// accesses per lane, then consume).  Per repetition: grid barrier (cg), then
// every warp times its 8 accesses with clock64; reported: mean and max per-warp
// latency (ns) averaged over repetitions.
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o mba tools/microbench_atomics.cu
#include <cooperative_groups.h>
#include <cstdio>
#include <cstdint>
#include <vector>

namespace cg = cooperative_groups;

template <int MODE>
__global__ void __launch_bounds__(512, 1) k_burst(unsigned long long *c64, uint32_t *c32,
                                                   const uint32_t *idx, int reps, int active_warps,
                                                   unsigned long long *out_sum,
                                                   unsigned long long *out_max) {
    cg::grid_group grid = cg::this_grid();
    const unsigned lane = threadIdx.x & 31;
    const unsigned gw = (blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    // round-robin: warp gw active iff its unit index < active_warps
    const unsigned unit = (threadIdx.x >> 5) * gridDim.x + blockIdx.x;
    for (int r = 0; r < reps; ++r) {
        grid.sync();
        if (unit < (unsigned)active_warps) {
            const uint32_t *ix = idx + ((size_t)(r % 16) * 4096 * 256) + (size_t)gw * 256 + lane;
            uint32_t w[8];
#pragma unroll
            for (int q = 0; q < 8; ++q) w[q] = ix[32 * q];
            const long long t0 = clock64();
            unsigned long long acc = 0;
            if (MODE == 0) {  // 64-bit atom.add with return
                unsigned long long o[8];
#pragma unroll
                for (int q = 0; q < 8; ++q)
                    asm volatile("atom.global.add.u64 %0, [%1], %2;" : "=l"(o[q]) : "l"(c64 + w[q]), "l"(~0ull));
#pragma unroll
                for (int q = 0; q < 8; ++q) acc += o[q];
            } else if (MODE == 1) {  // 32-bit atom.add with return
                uint32_t o[8];
#pragma unroll
                for (int q = 0; q < 8; ++q)
                    asm volatile("atom.global.add.u32 %0, [%1], %2;" : "=r"(o[q]) : "l"(c32 + w[q]), "r"(~0u));
#pragma unroll
                for (int q = 0; q < 8; ++q) acc += o[q];
            } else if (MODE == 2) {  // 64-bit plain loads
                unsigned long long o[8];
#pragma unroll
                for (int q = 0; q < 8; ++q) o[q] = __ldcg(c64 + w[q]);
#pragma unroll
                for (int q = 0; q < 8; ++q) acc += o[q];
            } else if (MODE == 4) {  // 32-bit atom.add on a 2x larger footprint (stride 2)
                uint32_t o[8];
#pragma unroll
                for (int q = 0; q < 8; ++q)
                    asm volatile("atom.global.add.u32 %0, [%1], %2;" : "=r"(o[q]) : "l"(reinterpret_cast<uint32_t *>(c64) + 2 * (size_t)w[q]), "r"(~0u));
#pragma unroll
                for (int q = 0; q < 8; ++q) acc += o[q];
            } else if (MODE == 5) {  // 64-bit atom.add on half the footprint
                unsigned long long o[8];
#pragma unroll
                for (int q = 0; q < 8; ++q)
                    asm volatile("atom.global.add.u64 %0, [%1], %2;" : "=l"(o[q]) : "l"(c64 + (w[q] >> 1)), "l"(~0ull));
#pragma unroll
                for (int q = 0; q < 8; ++q) acc += o[q];
            } else {  // contiguous 32-bit loads (a row segment): 8 x 128 B per warp
                const uint32_t *row = c32 + ((size_t)w[0] & ~1023ull);
                uint32_t o[8];
#pragma unroll
                for (int q = 0; q < 8; ++q) o[q] = __ldcs(row + 32 * q + lane);
#pragma unroll
                for (int q = 0; q < 8; ++q) acc += o[q];
            }
            const long long dt = clock64() - t0 + (acc == 12345 ? 1 : 0);
            const unsigned long long m = __reduce_max_sync(0xffffffffu, (unsigned)dt);
            if (lane == 0) {
                atomicAdd(out_sum, m);
                atomicMax(out_max + r, m);
            }
        }
    }
}

int main() {
    const size_t n = 16777216;
    unsigned long long *c64;
    uint32_t *c32, *idx;
    unsigned long long *sum, *mx;
    cudaMalloc(&c64, n * 8);
    cudaMalloc(&c32, n * 4);
    cudaMemset(c64, 0x7f, n * 8);
    cudaMemset(c32, 0x7f, n * 4);
    const size_t ni = (size_t)16 * 4096 * 256;
    std::vector<uint32_t> h(ni);
    uint64_t x = 88172645463325252ull;
    for (auto &v : h) {
        x ^= x << 13; x ^= x >> 7; x ^= x << 17;
        v = (uint32_t)(x % n);
    }
    cudaMalloc(&idx, ni * 4);
    cudaMemcpy(idx, h.data(), ni * 4, cudaMemcpyHostToDevice);
    const int reps = 400;
    cudaMalloc(&sum, 8);
    cudaMalloc(&mx, reps * 8);
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    int clk = 0;
    cudaDeviceGetAttribute(&clk, cudaDevAttrClockRate, 0);
    const char *names[6] = {"atom.add.u64 (ret) 134MB", "atom.add.u32 (ret) 67MB", "ld.u64 random 134MB",
                            "ld.u32 contiguous rows", "atom.add.u32 (ret) 134MB", "atom.add.u64 (ret) 67MB"};
    for (int mode = 0; mode < 6; ++mode) {
        for (int aw : {100, 800, 2368}) {
            cudaMemset(sum, 0, 8);
            cudaMemset(mx, 0, reps * 8);
            int active = aw;
            void *args[] = {&c64, &c32, &idx, (void *)&reps, &active, &sum, &mx};
            void *fn = mode == 0 ? (void *)k_burst<0> : mode == 1 ? (void *)k_burst<1>
                     : mode == 2 ? (void *)k_burst<2> : mode == 3 ? (void *)k_burst<3>
                     : mode == 4 ? (void *)k_burst<4> : (void *)k_burst<5>;
            cudaLaunchCooperativeKernel(fn, sms, 512, args, 0, 0);
            cudaError_t e = cudaDeviceSynchronize();
            unsigned long long hs = 0;
            std::vector<unsigned long long> hm(reps);
            cudaMemcpy(&hs, sum, 8, cudaMemcpyDeviceToHost);
            cudaMemcpy(hm.data(), mx, reps * 8, cudaMemcpyDeviceToHost);
            double mmax = 0;
            for (int r = 10; r < reps; ++r) mmax += hm[r];
            mmax /= (reps - 10);
            const double cyc_ns = 1e6 / clk;  // clk in kHz
            printf("%-28s warps %5d (x8 per lane = %7d accesses): mean warp %.0f ns, max warp %.0f ns  %s\n",
                   names[mode], aw, aw * 256, (double)hs / ((double)reps * aw) * cyc_ns, mmax * cyc_ns,
                   e == cudaSuccess ? "" : cudaGetErrorString(e));
        }
    }
    return 0;
}
