// gc_event.cu -- EVENT mode (work-efficient witness/resume sweep); see DESIGN.md.
#include "gc_internal.cuh"

namespace gc {

int run_event_maxmin(gc_graph *g, const RunParams &p, RunResult *r) {
    (void)g; (void)p; (void)r;
    set_error("GC_MODE_EVENT is not implemented yet");
    return GC_ERR_INVALID_ARG;
}

}  // namespace gc
