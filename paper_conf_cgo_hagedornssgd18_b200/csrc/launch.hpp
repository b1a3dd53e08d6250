// launch.hpp — host-side entry points of the kernel families (internal).
#pragma once
#include <cuda.h>
#include <cuda_runtime.h>

#include <cstdint>
#include <string>

#include "common.cuh"

namespace lift {

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

// K2T — two weighted 7-point steps per pass (temporal blocking), CLAMP/MIRROR/REFLECT.
bool sweep3d_t2_supported(const StencilParams& p);
cudaError_t launch_sweep3d_t2(const StencilParams& p, const float* in, float* out, cudaStream_t stream, int num_sms,
                              std::string* err);

// K1 — 2D TMA halo-tile kernel (weighted box r<=4, srad1, srad2).
bool tile2d_supported(const StencilParams& p);
cudaError_t launch_tile2d(const StencilParams& p, const float* in0, const float* in1, float* out,
                          cudaStream_t stream, int num_sms, std::string* err);

// OP_SRAD: q0^2 = var/mean^2 of the image (fp64, deterministic) into the
// workspace, as SRAD1's constants {q0, a, b}
size_t srad_workspace_bytes(int num_sms);
const float* srad_q0_ptr(void* ws, int num_sms);
cudaError_t launch_srad_q0(const float* img, int64_t n, void* ws, int num_sms, cudaStream_t stream);

// wait (one thread, acquire.sys) until *a >= value and *b >= value (NULL = skip)
cudaError_t launch_wait_signals(const unsigned int* a, const unsigned int* b, unsigned int value,
                                cudaStream_t stream);

}  // namespace lift
