// prune_f64_unit.cu -- FP64 F81 table kernels with the unit-diagonal branch loop (long
// alignments; prune_kernels.cuh, unit_branch), compiled beside prune_f64.cu.
#include "prune_kernels.cuh"

namespace mpcgs {
cudaError_t launch_tab_unit_f64(const PruneArgs& a, int ntrees, cudaStream_t st) {
    return launch_tab_dmx<double, PRUNE_SI64, true, false, 2, true>(a, ntrees, st);
}
}  // namespace mpcgs
