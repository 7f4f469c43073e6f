"""B200-native random-sampling rank-k approximation (Mary et al., SC15).

The compute path is the CUDA library ``lib/librs_lowrank.so`` (C ABI: ``include/rs_lowrank.h``);
``rs_lowrank`` is its thin Python binding.  PyTorch supplies device memory, streams and
process groups only.
"""

from . import rs_lowrank  # noqa: F401
from .rs_lowrank import (  # noqa: F401
    Qp3, RSError, create, destroy, kernel_launches, empty_colmajor, factor, get_fallbacks, get_info, get_pivot_data,
    get_profile, get_sample,
    load_library, omega, pivot, power_iterate, reset_profile, run, run_host, sample, sample_adaptive, set_profiling,
    qp3_truncated, sample_columns, set_sample,
    workspace_bytes,
)
