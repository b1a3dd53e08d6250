"""B200-native Lift stencil hot path (Hagedorn et al., CGO'18).

``map_n(f, slide_n(size, step, pad_n(l, r, h, input)))`` on
fp32 grids, run by hand-written sm_100a CUDA kernels in libstencil.so behind
the C ABI of include/stencil.h.  This package is the thin binding: ``_lib``
exposes the C functions under their C names, ``Plan`` wraps them for torch
tensors, ``slab`` adds the multi-GPU slab decomposition.
"""
from . import _lib
from ._lib import (StencilError, stencil_apply, stencil_apply_region, stencil_apply_region_put,  # noqa: F401
                   stencil_apply2_region,
                   stencil_iterate, stencil_slab_step_fused, stencil_wait_signals,
                   stencil_set_wait_timeout_ms, stencil_device_fault,
                   stencil_last_error, stencil_plan_create, stencil_plan_destroy,
                   stencil_plan_output_extents, stencil_plan_set_slab, stencil_plan_set_time_block,
                   stencil_plan_set_variant, stencil_plan_time_block,
                   stencil_plan_variant, stencil_plan_last_variant, stencil_plan_last_kernel,
                   stencil_plan_set_pad_decay,
                   stencil_run_host, stencil_run_host_batch, stencil_status_string,
                   stencil_version)
from .plan import Plan  # noqa: F401

__all__ = ["Plan", "StencilError"] + list(_lib.EXPORTED)
