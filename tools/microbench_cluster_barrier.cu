// Microbenchmark (tools/, not part of libgc): a grid barrier over one block per
// SM, flat (every block arrives on one word with a relaxed atomic and polls
// it) vs hierarchical through thread-block clusters (hardware cluster barrier,
// then one arrival and one poller per cluster, then the cluster barrier
// again).  Reports us per barrier.
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o mcb tools/microbench_cluster_barrier.cu
#include <cooperative_groups.h>
#include <cstdio>
namespace cg = cooperative_groups;

__device__ __forceinline__ unsigned long long ld_relaxed(const unsigned long long *p) {
    unsigned long long v;
    asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}

template <bool CLUSTER>
__global__ void k_bar(unsigned long long *word, int reps, unsigned nparties) {
    for (int r = 1; r <= reps; ++r) {
        if (CLUSTER) cg::this_cluster().sync();
        else __syncthreads();
        const bool leader = CLUSTER ? (cg::this_cluster().block_rank() == 0) : true;
        if (threadIdx.x == 0 && leader) {
            atomicAdd(word, 1ull);
            while (ld_relaxed(word) < (unsigned long long)nparties * r) {
            }
        }
        if (CLUSTER) cg::this_cluster().sync();
        else __syncthreads();
    }
}

int main() {
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    unsigned long long *w;
    cudaMalloc(&w, 8);
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    const int reps = 2000;
    for (int cs : {1, 2, 4, 8}) {
        cudaLaunchConfig_t cfg = {};
        cudaLaunchAttribute at[2];
        int na = 0;
        at[na].id = cudaLaunchAttributeCooperative;
        at[na].val.cooperative = 1;
        ++na;
        int blocks = sms;
        if (cs > 1) {
            at[na].id = cudaLaunchAttributeClusterDimension;
            at[na].val.clusterDim.x = cs;
            at[na].val.clusterDim.y = 1;
            at[na].val.clusterDim.z = 1;
            ++na;
            cfg.blockDim = dim3(768);
            cfg.gridDim = dim3(cs);
            cfg.attrs = at;
            cfg.numAttrs = na;
            int nclusters = 0;
            cudaOccupancyMaxActiveClusters(&nclusters, k_bar<true>, &cfg);
            blocks = (nclusters * cs) / cs * cs;
            if (blocks > sms) blocks = sms / cs * cs;
            printf("cluster %d: max active clusters %d -> %d blocks\n", cs, nclusters, blocks);
        }
        cfg.gridDim = dim3(blocks);
        cfg.blockDim = dim3(768);
        cfg.attrs = at;
        cfg.numAttrs = na;
        const unsigned parties = cs > 1 ? blocks / cs : blocks;
        cudaMemset(w, 0, 8);
        cudaError_t err;
        if (cs > 1) err = cudaLaunchKernelEx(&cfg, k_bar<true>, w, 10, parties);
        else err = cudaLaunchKernelEx(&cfg, k_bar<false>, w, 10, parties);
        cudaDeviceSynchronize();
        if (err != cudaSuccess) { printf("launch failed (cluster %d): %s\n", cs, cudaGetErrorString(err)); continue; }
        cudaMemset(w, 0, 8);
        cudaEventRecord(e0);
        if (cs > 1) cudaLaunchKernelEx(&cfg, k_bar<true>, w, reps, parties);
        else cudaLaunchKernelEx(&cfg, k_bar<false>, w, reps, parties);
        cudaEventRecord(e1);
        cudaEventSynchronize(e1);
        float ms = 0;
        cudaEventElapsedTime(&ms, e0, e1);
        printf("cluster size %d, %d blocks, %u arrivals: %.3f us per barrier (%s)\n", cs, blocks, parties,
               1e3 * ms / reps, cudaGetErrorString(cudaGetLastError()));
    }
    return 0;
}
