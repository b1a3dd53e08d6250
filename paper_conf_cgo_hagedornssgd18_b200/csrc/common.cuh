// common.cuh — launch parameters and index arithmetic shared by all kernels.
//
// The plan canonicalises every stencil to 3 dimensions (a 1D/2D grid gets
// leading dimensions of extent 1, size 1, step 1, pad 0), so every kernel
// indexes (z, y, x) with x contiguous.  Parameters travel by value as a
// __grid_constant__ struct: the plan owns no device memory and plans never
// share __constant__ symbols.
#pragma once
#include <cstdint>

#include <vector_types.h>

namespace lift {

enum PadKind : int { PAD_CLAMP = 0, PAD_MIRROR = 1, PAD_WRAP = 2, PAD_CONSTANT = 3, PAD_REFLECT = 4, PAD_DAMPEN = 5 };
enum OpKind : int {
  OP_WEIGHTED = 0, OP_HOTSPOT3D = 1, OP_SRAD1 = 2, OP_SRAD2 = 3, OP_ACOUSTIC = 4, OP_HOTSPOT2D = 5, OP_GRADIENT = 6,
  OP_SRAD = 7
};

constexpr int kMaxTaps = 125;     // 5x5x5
constexpr int kMaxParams = 16;
constexpr int kMaxInputs = 2;
constexpr int kMaxSep = 16;

struct StencilParams {
  // canonical 3D geometry (index 0 = z, slowest)
  int64_t n[3];          // owned input extents
  int64_t o[3];          // output extents
  int64_t row;           // elements per row (= n[2])
  int64_t plane;         // elements per plane (= n[1]*n[2])
  int32_t size[3], step[3], lo[3], hi[3];
  int32_t kind[3];
  float pad_value;
  float pad_decay;       // PAD_DAMPEN: factor per cell of distance outside the grid (reading A29)
  int32_t op;
  int32_t radius;        // star/box radius for non-WEIGHTED ops and fast kernels
  // slab mode along z (ghost == 0 and z_off == 0 and gnz == n[0] otherwise)
  int64_t z_off;         // global index of owned plane 0
  int64_t gnz;           // global extent of dimension 0
  int32_t ghost;         // ghost planes before/after the owned ones in every buffer
  int32_t slab;          // 1 when the plan is a slab of a larger grid
  // output region along dimension 0: [reg0, reg1)
  int64_t reg0, reg1;
  // WEIGHTED: non-zero taps in row-major window order
  int32_t ntaps;
  int16_t tap[kMaxTaps][3];   // window index k per dimension
  int32_t tap_off[kMaxTaps];   // kz*plane + ky*row + kx (K0 interior fast path; -1 in [0] = disabled)
  float w[kMaxTaps];
  float wbox[kMaxTaps];        // dense row-major window weights (fast kernels)
  // 2D WEIGHTED with exactly rank-1 weights w[ky][kx] = su[ky] * sv[kx]:
  // every kernel family evaluates sum_ky su[ky] * (sum_kx sv[kx] * x) in this order
  int32_t sep;
  float su[kMaxSep], sv[kMaxSep];
  float prm[kMaxParams];
  // fused halo put (slab mode, per launch): output plane z < ghost is also
  // stored at put_lo + z*plane, plane z >= n0 - ghost at put_hi + (z - (n0 -
  // ghost))*plane (the neighbours' ghost planes, NVLink peer pointers); the
  // last CTA then release-stores sig_value to sig_lo / sig_hi (system scope)
  float* put_lo;
  float* put_hi;
  unsigned int* sig_lo;
  unsigned int* sig_hi;
  unsigned int sig_value;
  // OP_SRAD (full iteration): device array {q0sqr, a, b} written by the q0
  // reduction before the stencil launch (SRAD1's constants, op_srad1)
  const float* srad_q0;
  // OP_SRAD, fused pass (K1S): q0 from srad_nparts fp64 (sum, sum of squares)
  // partials of the input image (reduced in-kernel, fixed order), and this
  // launch's own output statistics, one partial per CTA, into srad_part_out
  // (so the next iteration needs no reduction pass over I)
  const double2* srad_part_in;
  double2* srad_part_out;
  int32_t srad_nparts;
  // single-launch fused step: before loading ghost planes (first / last
  // z-chunk) the producer waits until *wait_lo / *wait_hi >= wait_value
  // (acquire, system scope); the boundary chunks are scheduled first and the
  // neighbours' flags are raised as soon as their chunk is complete
  const unsigned int* wait_lo;
  const unsigned int* wait_hi;
  unsigned int wait_value;
  int32_t fused_step;
  // bounded waits: give up after wait_timeout_ns (0 = never) and set the
  // fault word of the code (host-mapped block, read by stencil_device_fault)
  unsigned long long wait_timeout_ns;
  unsigned int* fault;
};

// fault codes of a timed-out wait: word fault[code - 1] of the host-visible
// fault block is set to 1
constexpr unsigned int kFaultWaitLo = 1u;   // flag of the lower neighbour never arrived
constexpr unsigned int kFaultWaitHi = 2u;   // flag of the upper neighbour never arrived

// h(i, n) of the reindexing pad (A1-A5).
// i is the unpadded index (padded index minus l).  Only called when i is out
// of [0, n).
__host__ __device__ __forceinline__ int64_t pad_remap(int64_t i, int64_t n, int kind) {
  switch (kind) {
    case PAD_CLAMP:
    case PAD_DAMPEN:     // the nearest element (scaled by the caller, dampen_pow)
      return i < 0 ? 0 : (i >= n ? n - 1 : i);
    case PAD_MIRROR: {
      if (i < 0) i = -1 - i;               // now i >= 0
      const int64_t p = 2 * n;
      i %= p;
      return i >= n ? p - 1 - i : i;
    }
    case PAD_WRAP: {
      i %= n;
      return i < 0 ? i + n : i;
    }
    case PAD_REFLECT: {
      if (n == 1) return 0;
      const int64_t p = 2 * n - 2;
      i %= p;
      if (i < 0) i += p;
      return i >= n ? p - i : i;
    }
    default:
      return i;
  }
}

// PAD_DAMPEN (reading A29): a cell d steps outside the grid holds the nearest
// element times decay^d, per dimension in pad_n's order, so a
// window element crossing k DAMPEN cells in total (over the dimensions inside
// the innermost out-of-range CONSTANT one) is x (or the constant) times
// decay^k — computed as a sequential product, identical in every kernel.
__host__ __device__ __forceinline__ int64_t outside_dist(int64_t i, int64_t n) {
  return i < 0 ? -i : (i >= n ? i - n + 1 : 0);
}
__device__ __forceinline__ float dampen_pow(float g, int64_t k) {
  float f = 1.0f;
  for (; k > 0; --k) f = __fmul_rn(f, g);
  return f;
}
__host__ __device__ __forceinline__ bool has_dampen(const StencilParams& p) {
  return p.kind[0] == PAD_DAMPEN || p.kind[1] == PAD_DAMPEN || p.kind[2] == PAD_DAMPEN;
}

// Local plane index (within a buffer of n0 + 2*ghost planes) of the input
// plane with GLOBAL index gz, or -1 when the padded value is the constant.
__host__ __device__ __forceinline__ int64_t plane_of(const StencilParams& p, int64_t gz) {
  if (gz < 0 || gz >= p.gnz) {
    if (p.kind[0] == PAD_CONSTANT) return -1;
    if (!(p.slab && p.kind[0] == PAD_WRAP)) gz = pad_remap(gz, p.gnz, p.kind[0]);
    // slab + wrap: ring neighbour's planes are in the ghosts
  }
  return gz - p.z_off + p.ghost;
}

// Programmatic dependent launch (sm_90+): a kernel launched with the
// programmatic-stream-serialization attribute may be scheduled while the
// previous kernel of the stream is still draining; it runs its prologue
// (mbarrier init, tensor-map prefetch), then waits here for the previous
// grid's completion and memory flush before touching global memory.  Both are
// no-ops for an ordinary launch.
__device__ __forceinline__ void pdl_wait() {
#if defined(__CUDA_ARCH__)
  asm volatile("griddepcontrol.wait;" ::: "memory");
#endif
}
__device__ __forceinline__ void pdl_launch_dependents() {
#if defined(__CUDA_ARCH__)
  asm volatile("griddepcontrol.launch_dependents;" ::: "memory");
#endif
}

}  // namespace lift
