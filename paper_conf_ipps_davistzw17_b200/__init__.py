"""B200-native hot path of the multiple-proposal coalescent genealogy sampler
(mpcgs; Davis 2016): one generalized Metropolis-Hastings step per device loop
iteration plus the theta MLE, as a C-ABI CUDA library (libmpcgs.so, sm_100a)
with a thin ctypes binding.  See DESIGN.md and include/mpcgs.h."""
from .mpcgs import (  # noqa: F401
    EXPORTS, MODELS, Context, MpcgsError, lib, mpcgs_nccl_unique_id, mpcgs_transition,
    mpcgs_sample_loci, mpcgs_estimate_theta_loci, mpcgs_em_loci, mpcgs_philox, mpcgs_phylip_read, mpcgs_parse_newick, mpcgs_prune_tiling, mpcgs_probe_peak,
    mpcgs_shard_range, mpcgs_tree_schedule, mpcgs_upgma, mpcgs_version, mpcgs_workspace_bytes, mpcgs_workspace_bytes_cfg,
)
