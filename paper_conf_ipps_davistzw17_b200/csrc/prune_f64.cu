// prune_f64.cu -- instantiates the pruning kernels for FP64 partials, F81 (Eq. 20).
#include "prune_kernels.cuh"

namespace mpcgs {
template cudaError_t launch_prune_typed<double, false>(PruneArgs, int, int, cudaStream_t, int&);
}  // namespace mpcgs
