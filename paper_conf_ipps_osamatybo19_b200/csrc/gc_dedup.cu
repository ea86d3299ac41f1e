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

#include <algorithm>
#include <cstdlib>
#include <vector>

#include "gc_internal.cuh"

namespace gc {

namespace {

// keep[ro[v]] = 1 for the first entry of every non-empty row v < n (absolute positions)
__global__ void k_row_start_marks(const int64_t *__restrict__ ro, int64_t n, uint8_t *mark) {
    for (int64_t v = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; v < n;
         v += (int64_t)gridDim.x * blockDim.x)
        if (ro[v + 1] > ro[v]) mark[ro[v]] = 1;
}

__global__ void k_keep(const uint32_t *__restrict__ ci, int64_t m, uint8_t *mark_keep) {
    for (int64_t e = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; e < m;
         e += (int64_t)gridDim.x * blockDim.x)
        mark_keep[e] = (mark_keep[e] || ci[e] != ci[e - 1]) ? 1 : 0;  // e == 0 is a row start (batch too)
}

__global__ void k_compact(const uint32_t *__restrict__ ci, const uint8_t *__restrict__ keep,
                          const uint32_t *__restrict__ pos, int64_t m, uint32_t *out) {
    for (int64_t e = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; e < m;
         e += (int64_t)gridDim.x * blockDim.x)
        if (keep[e]) out[pos[e]] = ci[e];
}

// new offsets of rows [0, n] of a batch whose entries start at e0 (m of
// them, batch-local positions pos / flags keep), kept entries before it: base
__global__ void k_new_offsets(const int64_t *__restrict__ ro, int64_t n, int64_t e0, int64_t m,
                              const uint32_t *__restrict__ pos, const uint8_t *__restrict__ keep,
                              int64_t base, int64_t *nro) {
    for (int64_t v = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; v <= n;
         v += (int64_t)gridDim.x * blockDim.x) {
        const int64_t e = ro[v] - e0;
        nro[v] = base + (e < m ? (int64_t)pos[e] : (m > 0 ? (int64_t)pos[m - 1] + keep[m - 1] : 0));
    }
}

struct RelOff {  // CUB offset iterator: absolute entry offset -> batch-relative (int)
    int64_t e0;
    __host__ __device__ __forceinline__ int64_t operator()(const int64_t &x) const { return x - e0; }
};

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
    return dedup_csr(g);  // sets g->deduped on success
}

// Rows are processed in batches of < 2^30 entries (CUB's int sizes; cfg5 has
// nnz > 2^31): per batch a segmented sort, the keep flags, an exclusive scan
// of them (batch-local positions) and the compaction at the running base.
int dedup_csr(gc_graph *g) {
    NvtxRange nv_("deduplicate CSR");
    const int64_t n = g->n, m = g->nnz;
    cudaStream_t st = g->stream;
    const int grid = g->sm_count * 8;
    int64_t kBatch = 1ll << 30;
    if (const char *b = std::getenv("GC_DEDUP_BATCH")) kBatch = std::max<long long>(1, std::atoll(b));  // test hook
    uint32_t *sorted = nullptr, *pos = nullptr, *nci = nullptr;
    uint8_t *keep = nullptr;
    int64_t *nro = nullptr;
    void *tmp = nullptr;
    size_t tmp_bytes = 0;
    int rc = GC_OK;
    cudaError_t e = cudaSuccess;
    std::vector<int64_t> h_ro((size_t)n + 1);
    int64_t base = 0;  // entries kept before the current batch
#define DD_TRY(expr, what)              \
    do {                                \
        e = (expr);                     \
        if (e != cudaSuccess) {         \
            rc = cuda_fail(e, what);    \
            goto out;                   \
        }                               \
    } while (0)
    if (cudaSuccess != dmalloc(&sorted, (size_t)std::max<int64_t>(m, 1) * 4) ||
        cudaSuccess != dmalloc(&pos, (size_t)std::max<int64_t>(m, 1) * 4) ||
        cudaSuccess != dmalloc(&keep, (size_t)std::max<int64_t>(m, 1)) ||
        cudaSuccess != dmalloc(&nci, (size_t)std::max<int64_t>(m, 1) * 4) ||
        cudaSuccess != dmalloc(&nro, (size_t)(n + 1) * 8)) {
        set_error("dedup: device allocation failed");
        rc = GC_ERR_OOM;
        goto out;
    }
    DD_TRY(cudaMemcpyAsync(h_ro.data(), g->ro, sizeof(int64_t) * (size_t)(n + 1), cudaMemcpyDeviceToHost, st),
           "dedup offsets");
    DD_TRY(cudaStreamSynchronize(st), "dedup offsets");
    if (m > 0) DD_TRY(cudaMemsetAsync(keep, 0, (size_t)m, st), "dedup marks");
    for (int64_t b0 = 0; b0 < n;) {
        // rows [b0, b1): as many as fit in kBatch entries (at least one row)
        int64_t b1 = b0 + 1;
        {
            int64_t lo = b0 + 1, hi = n;  // largest b1 with h_ro[b1] - h_ro[b0] <= kBatch
            while (lo < hi) {
                const int64_t mid = (lo + hi + 1) / 2;
                if (h_ro[mid] - h_ro[b0] <= kBatch) lo = mid;
                else hi = mid - 1;
            }
            b1 = lo;
        }
        const int64_t e0 = h_ro[b0], mb = h_ro[b1] - e0, nb = b1 - b0;
        if (mb >= (1ll << 31)) {
            set_error("dedup: a single row has more than 2^31 entries");
            rc = GC_ERR_TOO_LARGE;
            goto out;
        }
        if (mb > 0) {
            // CUB offsets relative to the batch's first entry
            auto rel = cub::TransformInputIterator<int64_t, RelOff, const int64_t *>(g->ro + b0, RelOff{e0});
            auto rel1 = cub::TransformInputIterator<int64_t, RelOff, const int64_t *>(g->ro + b0 + 1, RelOff{e0});
            size_t tb = 0, tb2 = 0;
            DD_TRY(cub::DeviceSegmentedSort::SortKeys(nullptr, tb, g->ci + e0, sorted + e0, (int)mb, (int)nb, rel,
                                                      rel1, st), "dedup sort");
            DD_TRY(cub::DeviceScan::ExclusiveSum(nullptr, tb2, keep + e0, pos + e0, (int)mb, st), "dedup scan");
            if (std::max(tb, tb2) > tmp_bytes) {
                dfree(tmp);
                tmp = nullptr;
                tmp_bytes = std::max(tb, tb2);
                if (cudaSuccess != dmalloc(&tmp, tmp_bytes + 16)) {
                    set_error("dedup: device allocation failed");
                    rc = GC_ERR_OOM;
                    goto out;
                }
            }
            DD_TRY(cub::DeviceSegmentedSort::SortKeys(tmp, tb, g->ci + e0, sorted + e0, (int)mb, (int)nb, rel,
                                                      rel1, st), "dedup sort");
            k_row_start_marks<<<grid, 256, 0, st>>>(g->ro + b0, nb, keep);
            k_keep<<<grid, 256, 0, st>>>(sorted + e0, mb, keep + e0);
            DD_TRY(cub::DeviceScan::ExclusiveSum(tmp, tb2, keep + e0, pos + e0, (int)mb, st), "dedup scan");
            k_compact<<<grid, 256, 0, st>>>(sorted + e0, keep + e0, pos + e0, mb, nci + base);
        }
        k_new_offsets<<<grid, 256, 0, st>>>(g->ro + b0, nb, e0, mb, pos + e0, keep + e0, base, nro + b0);
        DD_TRY(cudaGetLastError(), "dedup kernels");
        {
            int64_t kept = 0;  // nro[b1] = base + kept entries of the batch
            DD_TRY(cudaMemcpyAsync(&kept, nro + b1, 8, cudaMemcpyDeviceToHost, st), "dedup count");
            DD_TRY(cudaStreamSynchronize(st), "dedup count");
            base = kept;
        }
        b0 = b1;
    }
    if (n == 0) DD_TRY(cudaMemsetAsync(nro, 0, 8, st), "dedup offsets");
    DD_TRY(cudaStreamSynchronize(st), "dedup");
    if (g->owns_csr) {
        dfree(g->ro);
        dfree(g->ci);
    }
    g->ro = nro;
    g->ci = nci;
    g->nnz = base;
    g->owns_csr = true;
    g->deduped = true;
    dfree(g->s.deg);  // LDF degrees follow the rows
    g->s.deg = nullptr;
    nro = nullptr;
    nci = nullptr;
out:
#undef DD_TRY
    if (rc) cudaStreamSynchronize(st);  // queued kernels may still use the blocks
    dfree(sorted);
    dfree(pos);
    dfree(keep);
    dfree(nro);
    dfree(nci);
    dfree(tmp);
    return rc;
}

}  // namespace gc
