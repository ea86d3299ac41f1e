// gc_dist.cuh -- state of a partitioned graph (gc_dist.cu: sweep-based
// rounds; gc_dist_count.cu: COUNT-mode rounds).  Internal to libgc.
#pragma once

#include <vector>

#include "gc_internal.cuh"

#ifdef GC_HAVE_NCCL
#include <nccl.h>
#endif

namespace gc {

// COUNT-mode state of one partition (gc_dist_count.cu), allocated on first use
struct DCState {
    unsigned long long *cnt = nullptr;  // (hi << 32) | lo per owned vertex
    uint32_t *Z = nullptr;              // lo-freed-second stamps per owned vertex
    uint32_t *S = nullptr;              // scheduled owned vertices (monotone, | lo flag)
    void *L = nullptr;                  // long-row jobs of the round
    int64_t L_cap = 0;
    void *LC = nullptr;                 // their chunk items
    int64_t LC_cap = 0;
    int64_t *goff = nullptr;            // ghost rows: owned neighbours of each remote vertex,
    uint32_t *gadj = nullptr;           //   CSR over GLOBAL ids (empty for owned / non-neighbours)
    unsigned long long *ctr = nullptr;  // counters (gc_dist_count.cu)
    bool ghost_built = false;
};

struct Part {
    int64_t v0 = 0, v1 = 0, nnz = 0;
    int64_t *ro = nullptr;  // local offsets (start at 0)
    uint32_t *ci = nullptr; // global column ids
    bool owns_ro = false;
    uint32_t *C = nullptr;  // replicated colours [n_global]
    uint32_t *F[2] = {nullptr, nullptr};
    uint32_t *hub = nullptr;
    uint2 *colored = nullptr;  // pairs coloured this round [cap]
    uint2 *recv = nullptr;     // world * cap pairs
    unsigned long long *ctr = nullptr;
    unsigned long long *cnt_send = nullptr;  // [2]: coloured, remaining
    unsigned long long *cnt_recv = nullptr;  // [2 * world]
    int64_t *nk = nullptr;
    int64_t nk_cap = 1;
    DCState dc;
};

// Device-driven rounds (gc_dist_count.cu): every partition's
// inbox -- the coloured pairs the other partitions push to it each round and
// their per-round mailbox words.  Partition q's inbox lives in q's memory;
// on one GPU (loopback) all inboxes are local, across GPUs the other ranks'
// are mapped through CUDA IPC (NVLink peer access).
struct Inbox {
    uint2 *recv = nullptr;               // [2 slots][world sources][cap] pairs
    unsigned long long *mbox = nullptr;  // [2 slots][world sources] words
};

struct Dist {
    int64_t n_global = 0;
    int world = 1;
    int rank = 0;
    bool loopback = false;
    int64_t cap = 0;  // max vertices owned by any partition (pair padding)
    std::vector<Part> parts;
    unsigned long long *host_cnt = nullptr;  // pinned [2 * world]
#ifdef GC_HAVE_NCCL
    ncclComm_t comm = nullptr;
#endif
    // device-driven rounds: inboxes of all partitions (index = partition id)
    std::vector<Inbox> inbox;
    std::vector<void *> ipc_opened;      // peer mappings to close (multi-GPU)
    void *own_recv = nullptr, *own_mbox = nullptr;  // this rank's cudaMalloc'd inbox (multi-GPU)
    int persist_state = 0;               // 0 not set up, 1 ready, -1 unavailable (host rounds)
    uint32_t epoch = 0;                  // colourings run (mailbox tags)
};


int run_dist_count(gc_graph *g, const RunParams &p, RunResult *r, int64_t *frontier, int64_t fcap);
void free_inboxes(Dist &d);
void free_dist_count(Part &p);
int dist_reslice(gc_graph *g);  // after gc_dedup.cu replaced the handle's rows
int dist_exchange(gc_graph *g, size_t bytes, const std::vector<const void *> &send,
                  const std::vector<void *> &recv);
int nccl_fail(int e, const char *what);
int dist_wait(gc_graph *g);  // stream wait with NCCL async-error polling, timeout and abort

}  // namespace gc
