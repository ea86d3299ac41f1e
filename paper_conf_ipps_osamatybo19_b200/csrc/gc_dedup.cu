// gc_dedup.cu -- a deduplicated, row-sorted copy of the handle's CSR.
//
// The COUNT kernels need a symmetric adjacency MULTISET (a vertex's counts are
// decremented once per entry of its neighbours' rows).  Duplicate entries are
// legal input (the colouring depends on the adjacency SETS only, SURVEY 8(b),
// P:L719, R13); when a COUNT run reports an asymmetric multiset, the handle
// switches once to this copy (same sets, so the same colouring) and reruns.
// Per row: segmented sort (CUB), keep an entry iff it differs from its
// predecessor in the row, exclusive scan of the keep flags, compaction.
#include <cub/cub.cuh>

#include "gc_internal.cuh"

namespace gc {

namespace {

__global__ void k_row_start_marks(const int64_t *__restrict__ ro, int64_t n, uint8_t *mark) {
    for (int64_t v = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; v < n;
         v += (int64_t)gridDim.x * blockDim.x)
        if (ro[v + 1] > ro[v]) mark[ro[v]] = 1;
}

__global__ void k_keep(const uint32_t *__restrict__ ci, int64_t m, uint8_t *mark_keep) {
    for (int64_t e = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; e < m;
         e += (int64_t)gridDim.x * blockDim.x)
        mark_keep[e] = (mark_keep[e] || ci[e] != ci[e - 1]) ? 1 : 0;  // e == 0 is a row start
}

__global__ void k_compact(const uint32_t *__restrict__ ci, const uint8_t *__restrict__ keep,
                          const uint32_t *__restrict__ pos, int64_t m, uint32_t *out) {
    for (int64_t e = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; e < m;
         e += (int64_t)gridDim.x * blockDim.x)
        if (keep[e]) out[pos[e]] = ci[e];
}

__global__ void k_new_offsets(const int64_t *__restrict__ ro, int64_t n, int64_t m,
                              const uint32_t *__restrict__ pos, const uint8_t *__restrict__ keep,
                              int64_t *nro) {
    for (int64_t v = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; v <= n;
         v += (int64_t)gridDim.x * blockDim.x) {
        const int64_t e = ro[v];
        nro[v] = e < m ? (int64_t)pos[e] : (m > 0 ? (int64_t)pos[m - 1] + keep[m - 1] : 0);
    }
}

__global__ void k_rows_strict(const int64_t *__restrict__ ro, const uint32_t *__restrict__ ci,
                              int64_t n, unsigned int *bad) {
    for (int64_t v = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; v < n;
         v += (int64_t)gridDim.x * blockDim.x) {
        const int64_t e1 = ro[v + 1];
        for (int64_t e = ro[v] + 1; e < e1; ++e)
            if (ci[e] <= ci[e - 1]) {
                *bad = 1u;
                break;
            }
    }
}
}  // namespace

// Rows strictly increasing (no duplicates, sorted) -- checked once per handle.
// The JP kernels (Luby-MIS, Alg.2, Alg.4 in COUNT mode) need a duplicate-free
// adjacency before they start: a duplicate entry would be counted twice and
// JP has no safe asymmetry detection, so the handle switches to its
// deduplicated copy first when a row is not strictly increasing.
int ensure_strict_rows(gc_graph *g) {
    if (g->deduped || g->rows_strict) return GC_OK;
    unsigned int *bad = nullptr;
    unsigned int h = 0;
    GC_CUDA_TRY(dmalloc(&bad, 4));
    cudaError_t e = cudaMemsetAsync(bad, 0, 4, g->stream);
    if (e == cudaSuccess && g->n > 0) {
        k_rows_strict<<<g->sm_count * 8, 256, 0, g->stream>>>(g->ro, g->ci, g->n, bad);
        e = cudaGetLastError();
    }
    if (e == cudaSuccess) e = cudaMemcpyAsync(&h, bad, 4, cudaMemcpyDeviceToHost, g->stream);
    if (e == cudaSuccess) e = cudaStreamSynchronize(g->stream);
    dfree(bad);
    if (e != cudaSuccess) return cuda_fail(e, "row order check");
    if (!h) {
        g->rows_strict = true;
        return GC_OK;
    }
    g->deduped = true;
    return dedup_csr(g);
}

int dedup_csr(gc_graph *g) {
    const int64_t n = g->n, m = g->nnz;
    if (m >= (1ll << 31)) {
        set_error("dedup: more than 2^31 entries (the COUNT fallback copy is limited to int32 sizes)");
        return GC_ERR_TOO_LARGE;
    }
    cudaStream_t st = g->stream;
    const int grid = g->sm_count * 8;
    uint32_t *sorted = nullptr, *pos = nullptr, *nci = nullptr;
    uint8_t *keep = nullptr;
    int64_t *nro = nullptr;
    void *tmp = nullptr;
    size_t tb = 0, tb2 = 0;
    int rc = GC_OK;
    int64_t mm = 0;
    if (cudaSuccess != dmalloc(&sorted, (size_t)std::max<int64_t>(m, 1) * 4) ||
        cudaSuccess != dmalloc(&pos, (size_t)std::max<int64_t>(m, 1) * 4) ||
        cudaSuccess != dmalloc(&keep, (size_t)std::max<int64_t>(m, 1)) ||
        cudaSuccess != dmalloc(&nro, (size_t)(n + 1) * 8)) {
        rc = cuda_fail(cudaErrorMemoryAllocation, "dedup alloc");
        goto out;
    }
    if (m > 0) {
        GC_CUDA_TRY(cub::DeviceSegmentedSort::SortKeys(nullptr, tb, g->ci, sorted, (int)m, (int)n, g->ro,
                                                       g->ro + 1, st));
        GC_CUDA_TRY(cub::DeviceScan::ExclusiveSum(nullptr, tb2, keep, pos, (int)m, st));
        if (cudaSuccess != dmalloc(&tmp, std::max(tb, tb2) + 16)) {
            rc = cuda_fail(cudaErrorMemoryAllocation, "dedup temp");
            goto out;
        }
        GC_CUDA_TRY(cub::DeviceSegmentedSort::SortKeys(tmp, tb, g->ci, sorted, (int)m, (int)n, g->ro,
                                                       g->ro + 1, st));
        GC_CUDA_TRY(cudaMemsetAsync(keep, 0, (size_t)m, st));
        k_row_start_marks<<<grid, 256, 0, st>>>(g->ro, n, keep);
        k_keep<<<grid, 256, 0, st>>>(sorted, m, keep);
        GC_CUDA_TRY(cub::DeviceScan::ExclusiveSum(tmp, tb2, keep, pos, (int)m, st));
    }
    k_new_offsets<<<grid, 256, 0, st>>>(g->ro, n, m, pos, keep, nro);
    GC_CUDA_TRY(cudaGetLastError());
    GC_CUDA_TRY(cudaMemcpyAsync(&mm, nro + n, 8, cudaMemcpyDeviceToHost, st));
    GC_CUDA_TRY(cudaStreamSynchronize(st));
    if (cudaSuccess != dmalloc(&nci, (size_t)std::max<int64_t>(mm, 1) * 4)) {
        rc = cuda_fail(cudaErrorMemoryAllocation, "dedup output");
        goto out;
    }
    if (m > 0) k_compact<<<grid, 256, 0, st>>>(sorted, keep, pos, m, nci);
    GC_CUDA_TRY(cudaGetLastError());
    GC_CUDA_TRY(cudaStreamSynchronize(st));
    if (g->owns_csr) {
        dfree(g->ro);
        dfree(g->ci);
    }
    g->ro = nro;
    g->ci = nci;
    g->nnz = mm;
    g->owns_csr = true;
    nro = nullptr;
    nci = nullptr;
out:
    dfree(sorted);
    dfree(pos);
    dfree(keep);
    dfree(nro);
    dfree(nci);
    dfree(tmp);
    return rc;
}

}  // namespace gc
