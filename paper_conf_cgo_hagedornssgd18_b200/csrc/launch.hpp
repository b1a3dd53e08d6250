// launch.hpp — host-side entry points of the kernel families (internal).
#pragma once
#include <cuda.h>
#include <cuda_runtime.h>

#include <cstdint>
#include <cstdlib>
#include <string>

#include "common.cuh"

namespace lift {

// Whether stencil kernels are launched with programmatic dependent launch
// (overlaps a launch's ramp-up with the previous kernel's tail; every such
// kernel calls pdl_wait() before its first global access).  LIFT_PDL=0 turns
// it off (A/B measurement).
inline bool pdl_enabled() {
  static const bool on = [] {
    const char* e = getenv("LIFT_PDL");
    return !(e && e[0] == '0');
  }();
  return on;
}

// The kernel function the calling thread's most recent launch used (for
// stencil_plan_last_kernel: which kernel of a family ran, e.g. K2 or K2C).
inline thread_local const char* g_last_kernel = "none";
inline void set_last_kernel(const char* name) { g_last_kernel = name; }

inline cudaError_t launch_kernel(const void* fn, dim3 grid, dim3 block, void** args, size_t smem,
                                 cudaStream_t stream, bool pdl) {
  cudaLaunchConfig_t cfg{};
  cfg.gridDim = grid;
  cfg.blockDim = block;
  cfg.dynamicSmemBytes = smem;
  cfg.stream = stream;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
  at[0].val.programmaticStreamSerializationAllowed = (pdl && pdl_enabled()) ? 1 : 0;
  cfg.attrs = at;
  cfg.numAttrs = 1;
  return cudaLaunchKernelExC(&cfg, fn, args);
}

// K0 — generic remap kernel (any plan).
cudaError_t launch_generic(const StencilParams& p, const float* in0, const float* in1, float* out,
                           cudaStream_t stream, int num_sms);

// TMA tensor-map encoder (cuTensorMapEncodeTiled through the runtime's
// driver entry point; no -lcuda).  Returns false and sets ``err`` on failure.
bool encode_tensor_map_3d(CUtensorMap* map, const float* base, int64_t nx, int64_t ny, int64_t nz,
                          uint32_t box_x, uint32_t box_y, uint32_t box_z, std::string* err);

// K2 — 3D TMA plane-ring z-sweep (weighted star/box r<=2, hotspot3d, acoustic).
bool sweep3d_supported(const StencilParams& p);
cudaError_t launch_sweep3d(const StencilParams& p, const float* in0, const float* in1, float* out,
                           cudaStream_t stream, int num_sms, std::string* err);

// K2C — whole-column tiles for few-plane 3D grids (nz <= 16; radius-1 star
// weighted / Hotspot3D); launch_sweep3d routes eligible plans here.
bool column3d_supported(const StencilParams& p, const float* in0, const float* in1);
cudaError_t launch_column3d(const StencilParams& p, const float* in0, const float* in1, float* out,
                            cudaStream_t stream, std::string* err);

// K2CT — two steps per launch of a few-plane grid (Hotspot3D, reindexing
// pads): in0 = X_t, in1 = the point-wise grid, out = X_{t+2}.
bool column3d_t2_supported(const StencilParams& p, const float* in0, const float* in1);
cudaError_t launch_column3d_t2(const StencilParams& p, const float* in0, const float* in1, float* out,
                               cudaStream_t stream, std::string* err);

// K6 — all n steps of stencil_iterate for a few-plane 3D radius-1 star grid
// (weighted / Hotspot3D) with the grid resident in shared memory (one tile
// per SM, one cooperative launch, grid barrier per step).
bool resident3d_supported(const StencilParams& p, const float* s0, const float* s1, const float* aux,
                          int num_sms);
cudaError_t launch_resident3d(const StencilParams& p, float* s0, float* s1, const float* aux, int n_steps,
                              cudaStream_t stream, int num_sms, std::string* err);

// K2T — two weighted 7-point steps per pass (temporal blocking), CLAMP/MIRROR/REFLECT.
bool sweep3d_t2_supported(const StencilParams& p);
cudaError_t launch_sweep3d_t2(const StencilParams& p, const float* in, float* out, cudaStream_t stream, int num_sms,
                              std::string* err);

// K2R — two weighted 7-point steps per pass with X_{t+1} in registers
// (temporal blocking; x/y CLAMP/MIRROR/REFLECT, z CLAMP/MIRROR); the K2T
// entry point routes eligible plans here.
bool sweep3d_r2_supported(const StencilParams& p);
bool sweep3d_r2_auto(const StencilParams& p);          // the plans AUTO time blocking sends to K2R
cudaError_t launch_sweep3d_r2(const StencilParams& p, const float* in, float* out, cudaStream_t stream, int num_sms,
                              std::string* err);

// K2RA — two Acoustic (7 / 13-point, zero pad) steps per pass: reads u^{n-1}
// (prev) and u^n (cur), writes u^{n+1} (out1) and u^{n+2} (out2); four
// distinct buffers.
bool acoustic_r2_supported(const StencilParams& p);
bool acoustic_r2_auto(const StencilParams& p);        // the plans AUTO time blocking sends to K2RA
cudaError_t launch_acoustic_r2(const StencilParams& p, const float* prev, const float* cur, float* out1, float* out2,
                               cudaStream_t stream, int num_sms, std::string* err);

// K1 — 2D TMA halo-tile kernel (weighted box r<=4, srad1, srad2).
bool tile2d_supported(const StencilParams& p);
cudaError_t launch_tile2d(const StencilParams& p, const float* in0, const float* in1, float* out,
                          cudaStream_t stream, int num_sms, std::string* err);

// K3 — 2D per-warp TMA y-sweeps (the K1 ops; TMA-describable rows, x pad not WRAP).
bool wsweep2d_supported(const StencilParams& p, const float* in0, const float* in1, bool small);
cudaError_t launch_wsweep2d(const StencilParams& p, const float* in0, const float* in1, float* out,
                            cudaStream_t stream, int num_sms, std::string* err);

// OP_SRAD: q0^2 = var/mean^2 of the image (fp64, deterministic) into the
// workspace, as SRAD1's constants {q0, a, b}
size_t srad_workspace_bytes(int num_sms);
int srad_partials_cap(int num_sms);
double2* srad_partials_ptr(void* ws, int num_sms, int which);     // which = 0 / 1 (ping-pong)
const float* srad_q0_ptr(void* ws, int num_sms);
cudaError_t launch_srad_q0(const float* img, int64_t n, void* ws, int num_sms, cudaStream_t stream);
// (sum, sum of squares) partials of the image only (first iteration of a fused chain)
cudaError_t launch_srad_partials(const float* img, int64_t n, double2* partials, int num_sms, cudaStream_t stream,
                                 int* nparts);
// K1S: the fused SRAD pass; p.srad_part_in/srad_nparts/srad_part_out set;
// *nparts_out = partials written (one per CTA)
cudaError_t launch_srad_fused(const StencilParams& p, const float* in0, float* out, cudaStream_t stream,
                              int num_sms, std::string* err, int* nparts_out);

// K5 — WEIGHTED plans of any shape through shared-memory input boxes.
bool gather_supported(const StencilParams& p);
cudaError_t launch_gather(const StencilParams& p, const float* in0, float* out, cudaStream_t stream, int num_sms,
                          std::string* err);

// K4 — n steps of a small (L2-resident) 3D radius-1 star stencil (weighted
// star, Hotspot3D) in one persistent cooperative launch with grid barriers;
// the result is in s0 when n_steps is even, else in s1.
bool persist3d_supported(const StencilParams& p, const float* s0, const float* s1, const float* aux);
cudaError_t launch_persist3d(const StencilParams& p, float* s0, float* s1, const float* aux, int n_steps,
                             cudaStream_t stream, int num_sms, std::string* err);

// wait (one thread, acquire.sys) until *a >= value and *b >= value (NULL =
// skip); bounded by timeout_ns (0 = none), a timeout sets its fault word
cudaError_t launch_wait_signals(const unsigned int* a, const unsigned int* b, unsigned int value,
                                unsigned long long timeout_ns, unsigned int* fault, cudaStream_t stream);

}  // namespace lift
