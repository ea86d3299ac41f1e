// gc_dist.cu -- the colouring on a graph partitioned by contiguous vertex
// ranges: one partition per GPU (NCCL, one process per GPU),
// or P partitions inside one process on one GPU with a loopback transport of
// device copies (the same driver; used to test the partition / exchange logic
// bit-exactly on a single B200).
//
// Every partition owns rows [v0, v1) (column ids are global) and keeps a
// REPLICATED colour array C[n_global].  Round k of Alg.1/Alg.5 (P:L102-113,
// P:L506-556) on partition p:
//   1. sweep its uncoloured owned vertices against C (the round-start snapshot
//      for ghosts; owned colours are written in place, >= 2kH, which the status
//      test C[u] >= 2kH still counts as uncoloured: R6), publishing the
//      (vertex, colour) pairs coloured this round;
//   2. all-gather (newly coloured count, remaining count) of every partition;
//   3. all-gather the coloured pairs (padded to the largest count) and apply
//      the other partitions' pairs to C.
// After step 3 every replica equals the single-GPU C after round k, so the
// colouring is identical to the single-GPU one for any partition.  The loop
// stops when the summed remaining count is 0; every replica then holds all
// colours (no final gather needed).
#include <algorithm>
#include <cstring>
#include <chrono>
#include <cstdlib>
#include <thread>
#include <vector>

#include "gc_dist.cuh"

namespace gc {

int fill_u32(uint32_t *p, uint32_t val, int64_t n, cudaStream_t st);

// Wait for the handle's stream after NCCL work: polls the stream and the
// communicator's asynchronous error state; an NCCL error, or no progress for
// GC_NCCL_TIMEOUT_S seconds (default 120: a dead or hung peer), aborts the
// communicator (ncclCommAbort) and returns GC_ERR_NCCL instead of blocking
// forever in cudaStreamSynchronize.  The handle is unusable after an abort.
int dist_wait(gc_graph *g) {
    Dist &d = *g->dist;
#ifdef GC_HAVE_NCCL
    if (!d.loopback && d.comm) {
        double limit = 120.0;
        if (const char *e = std::getenv("GC_NCCL_TIMEOUT_S")) limit = std::max(1.0, std::atof(e));
        const auto t0 = std::chrono::steady_clock::now();
        for (unsigned spins = 0;; ++spins) {
            const cudaError_t q = cudaStreamQuery(g->stream);
            if (q == cudaSuccess) return GC_OK;
            if (q != cudaErrorNotReady) return cuda_fail(q, "distributed round");
            ncclResult_t ae = ncclSuccess;
            if (ncclCommGetAsyncError(d.comm, &ae) != ncclSuccess || ae != ncclSuccess) {
                ncclCommAbort(d.comm);
                d.comm = nullptr;
                return nccl_fail(ae, "asynchronous NCCL error (communicator aborted)");
            }
            if (std::chrono::duration<double>(std::chrono::steady_clock::now() - t0).count() > limit) {
                ncclCommAbort(d.comm);
                d.comm = nullptr;
                set_error("distributed round: no progress within GC_NCCL_TIMEOUT_S (peer dead or hung); "
                          "NCCL communicator aborted");
                return GC_ERR_NCCL;
            }
            if (spins > 64) std::this_thread::sleep_for(std::chrono::microseconds(20));
        }
    }
#endif
    GC_CUDA_TRY(cudaStreamSynchronize(g->stream));
    return GC_OK;
}

int nccl_fail(int e, const char *what) {
#ifdef GC_HAVE_NCCL
    std::string m = std::string("NCCL error in ") + what + ": " + ncclGetErrorString((ncclResult_t)e);
#else
    std::string m = std::string("NCCL unavailable (") + what + ")";
    (void)e;
#endif
    set_error(m);
    return GC_ERR_NCCL;
}

namespace {

__global__ void k_pack_counts(const unsigned long long *ctr, uint32_t k,
                              unsigned long long *cnt_send) {
    cnt_send[0] = ctr[kColoredCtr];
    cnt_send[1] = ctr[(k + 1) % 3];  // next frontier size
}

// Apply the coloured pairs received from the other partitions.
__global__ void k_apply(const uint2 *__restrict__ recv, const unsigned long long *cnt_recv,
                        int world, int self, int64_t stride, uint32_t *C) {
    for (int r = 0; r < world; ++r) {
        if (r == self) continue;
        const unsigned long long cnt = cnt_recv[2 * r];
        const uint2 *src = recv + (int64_t)r * stride;
        for (unsigned long long i = (unsigned long long)blockIdx.x * blockDim.x + threadIdx.x;
             i < cnt; i += (unsigned long long)gridDim.x * blockDim.x) {
            const uint2 pr = src[i];
            C[pr.x] = pr.y;
        }
    }
}

__global__ void k_rebase(const int64_t *ro, int64_t n_loc, int64_t *out) {
    const int64_t base = ro[0];
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i <= n_loc;
         i += (int64_t)gridDim.x * blockDim.x)
        out[i] = ro[i] - base;
}

int alloc_part(Part &p, int64_t n_global, int64_t cap, int world) {
    const int64_t nl = std::max<int64_t>(p.v1 - p.v0, 1);
    GC_CUDA_TRY(dmalloc(&p.C, sizeof(uint32_t) * (size_t)std::max<int64_t>(n_global, 1)));
    GC_CUDA_TRY(dmalloc(&p.F[0], sizeof(uint32_t) * (size_t)nl));
    GC_CUDA_TRY(dmalloc(&p.F[1], sizeof(uint32_t) * (size_t)nl));
    GC_CUDA_TRY(dmalloc(&p.hub, sizeof(uint32_t) * (size_t)nl));
    GC_CUDA_TRY(dmalloc(&p.colored, sizeof(uint2) * (size_t)std::max<int64_t>(cap, 1)));
    GC_CUDA_TRY(dmalloc(&p.recv, sizeof(uint2) * (size_t)std::max<int64_t>(cap, 1) * world));
    GC_CUDA_TRY(dmalloc(&p.ctr, 64 * sizeof(unsigned long long)));
    GC_CUDA_TRY(dmalloc(&p.cnt_send, 2 * sizeof(unsigned long long)));
    GC_CUDA_TRY(dmalloc(&p.cnt_recv, 2 * sizeof(unsigned long long) * world));
    GC_CUDA_TRY(dmalloc(&p.nk, sizeof(int64_t)));
    p.nk_cap = 1;
    return GC_OK;
}

void free_part(Part &p) {
    free_dist_count(p);
    if (p.owns_ro) dfree(p.ro);
    dfree(p.C);
    dfree(p.F[0]);
    dfree(p.F[1]);
    dfree(p.hub);
    dfree(p.colored);
    dfree(p.recv);
    dfree(p.ctr);
    dfree(p.cnt_send);
    dfree(p.cnt_recv);
    dfree(p.nk);
    p = Part();
}

// All-gather `bytes` from every partition's `send(p)` into `recv(p)`.
template <class SendF, class RecvF>
int exchange(gc_graph *g, size_t bytes, SendF send, RecvF recv) {
    Dist &d = *g->dist;
    if (bytes == 0) return GC_OK;
    if (d.loopback) {
        for (int p = 0; p < d.world; ++p)
            for (int q = 0; q < d.world; ++q)
                GC_CUDA_TRY(cudaMemcpyAsync((char *)recv(p) + (size_t)q * bytes, send(q), bytes,
                                            cudaMemcpyDeviceToDevice, g->stream));
        return GC_OK;
    }
#ifdef GC_HAVE_NCCL
    ncclResult_t e = ncclAllGather(send(0), recv(0), bytes, ncclUint8, d.comm, g->stream);
    if (e != ncclSuccess) return nccl_fail(e, "ncclAllGather");
    return GC_OK;
#else
    return nccl_fail(0, "exchange");
#endif
}

}  // namespace

// The handle's rows were replaced by their deduplicated copy (gc_dedup.cu):
// point every partition at its rows of the new CSR and drop its COUNT state
// (ghost rows and list capacities follow the rows).
int dist_reslice(gc_graph *g) {
    Dist &d = *g->dist;
    if (!d.loopback) {
        Part &p = d.parts[0];
        p.ro = g->ro;
        p.ci = g->ci;
        p.nnz = g->nnz;
        free_dist_count(p);
        return GC_OK;
    }
    std::vector<int64_t> h_ro((size_t)d.n_global + 1);
    GC_CUDA_TRY(cudaMemcpyAsync(h_ro.data(), g->ro, sizeof(int64_t) * h_ro.size(), cudaMemcpyDeviceToHost,
                                g->stream));
    GC_CUDA_TRY(cudaStreamSynchronize(g->stream));
    for (Part &p : d.parts) {
        p.nnz = h_ro[p.v1] - h_ro[p.v0];
        p.ci = g->ci + h_ro[p.v0];
        k_rebase<<<64, 256, 0, g->stream>>>(g->ro + p.v0, p.v1 - p.v0, p.ro);
        free_dist_count(p);
    }
    GC_CUDA_TRY(cudaGetLastError());
    return GC_OK;
}


int dist_exchange(gc_graph *g, size_t bytes, const std::vector<const void *> &send,
                  const std::vector<void *> &recv) {
    return exchange(g, bytes, [&](int q) { return send[q]; }, [&](int q) { return recv[q]; });
}

void destroy_dist(gc_graph *g) {
    if (!g || !g->dist) return;
    Dist &d = *g->dist;
    cudaDeviceSynchronize();  // the inboxes may be peer-mapped: no pending work may use them
    free_inboxes(d);
    for (auto &p : d.parts) free_part(p);
    if (d.host_cnt) hfree(d.host_cnt);
#ifdef GC_HAVE_NCCL
    if (d.comm) ncclCommDestroy(d.comm);
#endif
    delete g->dist;
    g->dist = nullptr;
}

// The colouring loop over all partitions of the handle.
int run_dist(gc_graph *g, const RunParams &p, RunResult *r, int64_t *frontier, int64_t fcap) {
    Dist &d = *g->dist;
    const int64_t n = d.n_global;
    r->rounds = r->inner = r->launches = 0;
    for (auto &pt : d.parts) {
        int rc = fill_u32(pt.C, GC_UNC, n, g->stream);
        if (rc) return rc;
        GC_CUDA_TRY(cudaMemsetAsync(pt.ctr, 0, 64 * sizeof(unsigned long long), g->stream));
    }
    const int64_t blocks_hub = g->sm_count * 2;
    int64_t k = 0;
    int64_t remaining = n;
    while (remaining > 0) {
        if (k >= p.max_rounds) {
            set_error("distributed colouring exceeded the round limit");
            return GC_ERR_TOO_LARGE;
        }
        if (frontier && k < fcap) frontier[k] = remaining;
        for (auto &pt : d.parts) {
            const int64_t nl = pt.v1 - pt.v0;
            GC_CUDA_TRY(cudaMemsetAsync(pt.ctr + kColoredCtr, 0, sizeof(unsigned long long), g->stream));
            SweepArgs a;
            a.ro = pt.ro;
            a.ci = pt.ci;
            a.C = pt.C;
            a.Fin = pt.F[k & 1];
            a.Fout = pt.F[(k + 1) & 1];
            a.hub = pt.hub;
            a.ctr = pt.ctr;
            a.nk = pt.nk;
            a.nk_cap = 0;
            a.k = (uint32_t)k;
            a.H = p.H;
            a.keys = p.keys;
            a.dense = k == 0 ? 1 : 0;
            a.n_loc = nl;
            a.v0 = (uint32_t)pt.v0;
            a.thread_max = (uint32_t)p.thread_deg_max;
            a.hub_min = (uint32_t)p.hub_deg_min;
            a.colored = pt.colored;
            const int blocks = (int)std::max<int64_t>(
                1, std::min<int64_t>((nl + 255) / 256, (int64_t)g->sm_count * 8));
            int rc = sweep_round(a, g->stream, blocks, (int)blocks_hub);
            if (rc) return rc;
            k_pack_counts<<<1, 1, 0, g->stream>>>(pt.ctr, (uint32_t)k, pt.cnt_send);
            r->launches += 3;
        }
        int rc = exchange(g, 2 * sizeof(unsigned long long),
                          [&](int q) { return (const void *)d.parts[q].cnt_send; },
                          [&](int q) { return (void *)d.parts[q].cnt_recv; });
        if (rc) return rc;
        GC_CUDA_TRY(cudaMemcpyAsync(d.host_cnt, d.parts[0].cnt_recv,
                                    2 * sizeof(unsigned long long) * d.world,
                                    cudaMemcpyDeviceToHost, g->stream));
        if ((rc = dist_wait(g))) return rc;
        unsigned long long maxc = 0, rem = 0;
        for (int q = 0; q < d.world; ++q) {
            maxc = std::max(maxc, d.host_cnt[2 * q]);
            rem += d.host_cnt[2 * q + 1];
        }
        if (maxc > (unsigned long long)d.cap) {
            set_error("internal: coloured pairs exceed the partition capacity");
            return GC_ERR_CUDA;
        }
        if (maxc > 0) {
            rc = exchange(g, sizeof(uint2) * maxc,
                          [&](int q) { return (const void *)d.parts[q].colored; },
                          [&](int q) { return (void *)d.parts[q].recv; });
            if (rc) return rc;
            for (size_t q = 0; q < d.parts.size(); ++q) {
                const int self = d.loopback ? (int)q : d.rank;
                k_apply<<<g->sm_count * 4, 256, 0, g->stream>>>(d.parts[q].recv, d.parts[q].cnt_recv,
                                                                d.world, self, (int64_t)maxc,
                                                                d.parts[q].C);
                r->launches += 1;
            }
        }
        GC_CUDA_TRY(cudaGetLastError());
        remaining = (int64_t)rem;
        ++k;
    }
    r->rounds = k;
    r->inner = k;
    return GC_OK;
}

}  // namespace gc

using namespace gc;

extern "C" {

int gc_nccl_unique_id(void *out128) {
    if (!out128) {
        set_error("gc_nccl_unique_id: NULL");
        return GC_ERR_INVALID_ARG;
    }
#ifdef GC_HAVE_NCCL
    static_assert(sizeof(ncclUniqueId) == 128, "ncclUniqueId is 128 bytes");
    ncclUniqueId id;
    ncclResult_t e = ncclGetUniqueId(&id);
    if (e != ncclSuccess) return nccl_fail(e, "ncclGetUniqueId");
    memcpy(out128, &id, 128);
    return GC_OK;
#else
    return nccl_fail(0, "gc_nccl_unique_id");
#endif
}

int gc_create_csr_internal(int64_t n, int64_t nnz, const int64_t *row_offsets,
                           const uint32_t *col_indices, uint32_t flags, gc_graph **out,
                           int64_t v_begin, int64_t n_global);

int gc_create_csr_dist(int64_t n_global, int64_t v_begin, int64_t v_end, int64_t nnz_local,
                       const int64_t *row_offsets_local, const uint32_t *col_indices_global,
                       const void *nccl_unique_id, int rank, int world, uint32_t flags,
                       gc_graph **out) {
    if (out) *out = nullptr;
    if (!out || !nccl_unique_id || world < 1 || rank < 0 || rank >= world || v_begin < 0 ||
        v_end < v_begin || v_end > n_global) {
        set_error("gc_create_csr_dist: bad arguments");
        return GC_ERR_INVALID_ARG;
    }
#ifndef GC_HAVE_NCCL
    set_error("gc_create_csr_dist: libgc was built without NCCL");
    return GC_ERR_NCCL;
#else
    gc_graph *g = nullptr;
    int rc = gc_create_csr_internal(v_end - v_begin, nnz_local, row_offsets_local,
                                    col_indices_global, flags, &g, v_begin, n_global);
    if (rc) return rc;
    g->dist = new Dist();
    Dist &d = *g->dist;
    d.n_global = n_global;
    d.world = world;
    d.rank = rank;
    d.loopback = false;
    ncclUniqueId id;
    memcpy(&id, nccl_unique_id, 128);
    ncclResult_t e = ncclCommInitRank(&d.comm, world, id, rank);
    if (e != ncclSuccess) {
        gc_destroy(g);
        return nccl_fail(e, "ncclCommInitRank");
    }
    // padding capacity: the largest owned range over all ranks
    unsigned long long *tmp = nullptr;
    unsigned long long mine = (unsigned long long)(v_end - v_begin), mx = 0;
    cudaError_t ce = dmalloc(&tmp, sizeof(unsigned long long));
    if (ce == cudaSuccess) ce = cudaMemcpy(tmp, &mine, sizeof(mine), cudaMemcpyHostToDevice);
    if (ce != cudaSuccess) {
        dfree(tmp);
        gc_destroy(g);
        return cuda_fail(ce, "dist setup");
    }
    e = ncclAllReduce(tmp, tmp, 1, ncclUint64, ncclMax, d.comm, 0);
    if (e == ncclSuccess) ce = cudaMemcpy(&mx, tmp, sizeof(mx), cudaMemcpyDeviceToHost);
    dfree(tmp);
    if (e != ncclSuccess || ce != cudaSuccess) {
        gc_destroy(g);
        return e != ncclSuccess ? nccl_fail(e, "ncclAllReduce") : cuda_fail(ce, "dist setup");
    }
    d.cap = (int64_t)mx;
    d.parts.resize(1);
    Part &p = d.parts[0];
    p.v0 = v_begin;
    p.v1 = v_end;
    p.nnz = nnz_local;
    p.ro = g->ro;
    p.ci = g->ci;
    p.owns_ro = false;
    rc = alloc_part(p, n_global, d.cap, world);
    if (rc == GC_OK && hmalloc(&d.host_cnt, 2 * sizeof(unsigned long long) * world) != cudaSuccess)
        rc = GC_ERR_OOM;
    if (rc) {
        gc_destroy(g);
        return rc;
    }
    *out = g;
    return GC_OK;
#endif
}

int gc_create_csr_loopback(int64_t n, int64_t nnz, const int64_t *row_offsets,
                           const uint32_t *col_indices, int parts, uint32_t flags,
                           gc_graph **out) {
    if (out) *out = nullptr;
    if (!out || parts < 1 || parts > 1024 || n < 0) {
        set_error("gc_create_csr_loopback: bad arguments");
        return GC_ERR_INVALID_ARG;
    }
    gc_graph *g = nullptr;
    int rc = gc_create_csr_internal(n, nnz, row_offsets, col_indices, flags, &g, 0, n);
    if (rc) return rc;
    g->dist = new Dist();
    Dist &d = *g->dist;
    d.n_global = n;
    d.world = parts;
    d.loopback = true;
    const int64_t chunk = (n + parts - 1) / parts;
    d.cap = std::max<int64_t>(chunk, 1);
    d.parts.resize(parts);
    std::vector<int64_t> h_ro(n + 1);
    cudaError_t ce = cudaMemcpy(h_ro.data(), g->ro, sizeof(int64_t) * (size_t)(n + 1),
                                cudaMemcpyDeviceToHost);
    if (ce != cudaSuccess) {
        gc_destroy(g);
        return cuda_fail(ce, "loopback setup");
    }
    for (int q = 0; q < parts; ++q) {
        Part &p = d.parts[q];
        p.v0 = std::min<int64_t>(n, (int64_t)q * chunk);
        p.v1 = std::min<int64_t>(n, p.v0 + chunk);
        p.nnz = h_ro[p.v1] - h_ro[p.v0];
        p.ci = g->ci + h_ro[p.v0];
        ce = dmalloc(&p.ro, sizeof(int64_t) * (size_t)(p.v1 - p.v0 + 1));
        if (ce != cudaSuccess) {
            gc_destroy(g);
            return cuda_fail(ce, "loopback setup");
        }
        p.owns_ro = true;
        k_rebase<<<64, 256>>>(g->ro + p.v0, p.v1 - p.v0, p.ro);
        rc = alloc_part(p, n, d.cap, parts);
        if (rc) {
            gc_destroy(g);
            return rc;
        }
    }
    if (hmalloc(&d.host_cnt, 2 * sizeof(unsigned long long) * parts) != cudaSuccess) {
        gc_destroy(g);
        return GC_ERR_OOM;
    }
    ce = cudaDeviceSynchronize();
    if (ce != cudaSuccess) {
        gc_destroy(g);
        return cuda_fail(ce, "loopback setup");
    }
    *out = g;
    return GC_OK;
}

int64_t gc_color_dist(gc_graph *g, const gc_options *o, int32_t *colors_out, gc_stats *stats) {
    Dist &d = *g->dist;
    const int kind = GC_VARIANT_KIND(o->variant);
    if (kind == GC_LUBY_MIS || kind == GC_IS_ALG2 || kind == GC_JP_ALG4 || kind == GC_HASH_IS(0)) {
        set_error("distributed colouring supports GC_MAXMIN and GC_MULTIHASH(h)");
        return GC_ERR_INVALID_ARG;
    }
    const int H = kind == GC_MULTIHASH(0) ? GC_VARIANT_HASHES(o->variant) : 1;
    RunParams p;
    p.H = H;
    for (int j = 0; j < H; ++j) p.keys.k[j] = weight_key(o->seed, j);
    p.thread_deg_max = o->thread_deg_max > 0 ? o->thread_deg_max : 8;
    p.hub_deg_min = o->hub_deg_min > 0 ? o->hub_deg_min : 4096;
    p.max_rounds = (int64_t)(0x7FFFFFFFll / (2 * H)) + 1;
    Profile prof;
    prof.on = (o->flags & GC_PROFILE) != 0;
    p.prof = &prof;
    int rc = ensure_scratch(g, false, false);
    if (rc) return rc;
    cudaEvent_t e0, e1;
    GC_CUDA_TRY(cudaEventCreate(&e0));
    GC_CUDA_TRY(cudaEventCreate(&e1));
    GC_CUDA_TRY(cudaEventRecord(e0, g->stream));
    RunResult res;
    int64_t *fs = stats ? stats->frontier_sizes : nullptr;
    const int64_t fcap = stats ? stats->frontier_cap : 0;
    // max-min: COUNT rounds (gc_dist_count.cu) unless SWEEP is asked for;
    // multi-hash: the sweep rounds
    const int mode_used = (H == 1 && o->mode != GC_MODE_SWEEP) ? GC_MODE_COUNT : GC_MODE_SWEEP;
    if (mode_used == GC_MODE_COUNT)
        rc = run_dist_count(g, p, &res, fs, fcap);
    else
        rc = run_dist(g, p, &res, fs, fcap);
    if (rc) {
        cudaEventDestroy(e0);
        cudaEventDestroy(e1);
        return rc;
    }
    // every replica holds all colours: count / compact / copy out of partition 0
    uint32_t *C = d.parts[0].C;
    int64_t launches = res.launches;
    const int64_t ncol = count_colors_device(g, C, d.n_global, (o->flags & GC_COMPACT) != 0, C,
                                             &launches);
    if (ncol < 0) return ncol;
    if (d.n_global > 0) {
        if (o->flags & GC_OUT_LOCAL_SLICE) {
            const Part &me = d.parts[0];
            GC_CUDA_TRY(cudaMemcpyAsync(colors_out, C + (d.loopback ? 0 : me.v0),
                                        sizeof(int32_t) * (size_t)(d.loopback ? d.n_global
                                                                              : me.v1 - me.v0),
                                        cudaMemcpyDefault, g->stream));
        } else {
            GC_CUDA_TRY(cudaMemcpyAsync(colors_out, C, sizeof(int32_t) * (size_t)d.n_global,
                                        cudaMemcpyDefault, g->stream));
        }
    }
    GC_CUDA_TRY(cudaEventRecord(e1, g->stream));
    GC_CUDA_TRY(cudaEventSynchronize(e1));
    float ms = 0.f;
    cudaEventElapsedTime(&ms, e0, e1);
    cudaEventDestroy(e0);
    cudaEventDestroy(e1);
    if ((o->flags & GC_COMPACT) == 0 && (uint64_t)2 * (uint64_t)res.rounds * (uint64_t)H > 0x7FFFFFFFull) {
        set_error("colours exceed INT32_MAX; use GC_COMPACT");
        return GC_ERR_TOO_LARGE;
    }
    if (stats) {
        stats->mode_used = mode_used;
        for (int c = 0; c < 4; ++c) {
            stats->kernel_ms[c] = prof.ms[c];
            stats->kernel_launches[c] = prof.launches[c];
            stats->kernel_bytes[c] = prof.bytes[c];
        }
        stats->visits = prof.visits;
        stats->rounds = res.rounds;
        stats->inner_iterations = res.inner;
        stats->n_colors = ncol;
        stats->launches = launches;
        stats->ms = ms;
    }
    return ncol;
}

}  // extern "C"
