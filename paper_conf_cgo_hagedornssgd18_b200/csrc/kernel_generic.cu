// kernel_generic.cu — K0: the generic remap kernel.
//
// One thread per output point (grid-stride).  Every tap is read straight from
// global memory at the padded index o*step + k (slide), remapped by
// h or replaced by the constant when it falls outside the grid (pad,
// P:407-466) — the "view" of P:880-893: nothing is copied.  K0 runs any plan
// (any ndim <= 3, size, step, pad, kind, op); it is the correctness baseline
// and the fallback for shapes the TMA kernels do not take (unaligned pointers,
// nx % 4 != 0, step > 1, 1D, wide windows).
#include <cuda_runtime.h>

#include "common.cuh"
#include "launch.hpp"
#include "ops.cuh"

namespace lift {
namespace {

struct Geo {
  int64_t oz, oy, ox;
};

// padded-grid read for one input: window element at unpadded coordinates
// (gz global plane, iy, ix).  Dimensions resolve innermost first (pad_n pads
// the outer dimension first, so an inner pad sees the outer one's
// cells): a CONSTANT dimension out of range gives the value, DAMPEN counts
// its distance (reading A29), the others remap.
__device__ __forceinline__ float fetch(const StencilParams& p, const float* __restrict__ in,
                                       int64_t gz, int64_t iy, int64_t ix) {
  int64_t nd = 0;
  if (ix < 0 || ix >= p.n[2]) {
    if (p.kind[2] == PAD_CONSTANT) return p.pad_value;
    if (p.kind[2] == PAD_DAMPEN) nd += outside_dist(ix, p.n[2]);
    ix = pad_remap(ix, p.n[2], p.kind[2]);
  }
  if (iy < 0 || iy >= p.n[1]) {
    if (p.kind[1] == PAD_CONSTANT) return nd ? __fmul_rn(p.pad_value, dampen_pow(p.pad_decay, nd)) : p.pad_value;
    if (p.kind[1] == PAD_DAMPEN) nd += outside_dist(iy, p.n[1]);
    iy = pad_remap(iy, p.n[1], p.kind[1]);
  }
  if (p.kind[0] == PAD_DAMPEN) nd += outside_dist(gz, p.gnz);
  const int64_t lz = plane_of(p, gz);
  const float v = lz < 0 ? p.pad_value : __ldg(in + lz * p.plane + iy * p.row + ix);
  return nd ? __fmul_rn(v, dampen_pow(p.pad_decay, nd)) : v;
}

// Accessor for centred ops: at<DZ,DY,DX>() is the window element at offset D
// from the window centre c_d = (size_d - 1) / 2.
struct CentredAcc {
  const StencilParams& p;
  const float* __restrict__ in;
  Geo g;
  template <int DZ, int DY, int DX>
  __device__ __forceinline__ float at() const {
    const int64_t gz = p.z_off + g.oz * p.step[0] + (p.size[0] - 1) / 2 + DZ - p.lo[0];
    const int64_t iy = g.oy * p.step[1] + (p.size[1] - 1) / 2 + DY - p.lo[1];
    const int64_t ix = g.ox * p.step[2] + (p.size[2] - 1) / 2 + DX - p.lo[2];
    return fetch(p, in, gz, iy, ix);
  }
};

// OP_SRAD: the diffusion coefficient c = SRAD1(I) at the padded position
// (oy + DY, ox + DX) — c is read through the plan's pad like any grid (A27)
struct SradCAcc {
  const StencilParams& p;
  const float* __restrict__ in;
  Geo g;
  template <int DZ, int DY, int DX>
  __device__ __forceinline__ float at() const {
    int64_t cy = g.oy + DY, cx = g.ox + DX;
    if (cy < 0 || cy >= p.n[1]) cy = pad_remap(cy, p.n[1], p.kind[1]);
    if (cx < 0 || cx >= p.n[2]) cx = pad_remap(cx, p.n[2], p.kind[2]);
    return op_srad1(CentredAcc{p, in, Geo{g.oz, cy, cx}}, p.srad_q0);
  }
};

__global__ void __launch_bounds__(256) k0_generic(const __grid_constant__ StencilParams p,
                                                  const float* __restrict__ in0,
                                                  const float* __restrict__ in1,
                                                  float* __restrict__ out) {
  pdl_launch_dependents();
  pdl_wait();
  const int64_t o1 = p.o[1], o2 = p.o[2];
  const int64_t per_plane = o1 * o2;
  const int64_t total = (p.reg1 - p.reg0) * per_plane;
  const int64_t out_plane = p.o[1] * p.o[2];
  for (int64_t idx = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; idx < total;
       idx += (int64_t)gridDim.x * blockDim.x) {
    Geo g;
    g.oz = p.reg0 + idx / per_plane;
    const int64_t rem = idx % per_plane;
    g.oy = rem / o2;
    g.ox = rem % o2;
    float v;
    switch (p.op) {
      case OP_WEIGHTED: {
        float acc = 0.0f;
        const int64_t bz = p.z_off + g.oz * p.step[0] - p.lo[0];
        const int64_t by = g.oy * p.step[1] - p.lo[1];
        const int64_t bx = g.ox * p.step[2] - p.lo[2];
        if (p.sep) {
          // separable 2D weights: rows first (x taps in order), then the column
          for (int ky = 0; ky < p.size[1]; ++ky) {
            float h = 0.0f;
            for (int kx = 0; kx < p.size[2]; ++kx) h = __fmaf_rn(p.sv[kx], fetch(p, in0, bz, by + ky, bx + kx), h);
            acc = __fmaf_rn(p.su[ky], h, acc);
          }
        } else {
          // interior fast path: the whole window lies inside the grid (and, in
          // slab mode, inside the global domain), so no tap needs a remap
          const bool inside = p.tap_off[0] >= 0 && bz >= 0 && bz + p.size[0] <= p.gnz && by >= 0 &&
                              by + p.size[1] <= p.n[1] && bx >= 0 && bx + p.size[2] <= p.n[2];
          if (inside) {
            const float* __restrict__ base = in0 + (bz - p.z_off + p.ghost) * p.plane + by * p.row + bx;
            for (int t = 0; t < p.ntaps; ++t) acc = __fmaf_rn(p.w[t], __ldg(base + p.tap_off[t]), acc);
          } else {
            for (int t = 0; t < p.ntaps; ++t) {
              const float x = fetch(p, in0, bz + p.tap[t][0], by + p.tap[t][1], bx + p.tap[t][2]);
              acc = __fmaf_rn(p.w[t], x, acc);
            }
          }
        }
        v = acc;
        break;
      }
      case OP_HOTSPOT3D: {
        const float Pc = __ldg(in1 + (g.oz + p.ghost) * p.plane + g.oy * p.row + g.ox);
        v = op_hotspot3d(CentredAcc{p, in0, g}, Pc, p.prm);
        break;
      }
      case OP_SRAD1:
        v = op_srad1(CentredAcc{p, in0, g}, p.prm);
        break;
      case OP_SRAD2:
        v = op_srad2(CentredAcc{p, in0, g}, CentredAcc{p, in1, g}, p.prm);
        break;
      case OP_HOTSPOT2D:
        v = op_hotspot2d(CentredAcc{p, in0, g}, CentredAcc{p, in1, g}, p.prm);
        break;
      case OP_GRADIENT:
        v = op_gradient(CentredAcc{p, in0, g}, p.prm);
        break;
      case OP_SRAD:
        v = op_srad2(SradCAcc{p, in0, g}, CentredAcc{p, in0, g}, p.prm);
        break;
      case OP_ACOUSTIC: {
        // inputs: in0 = prev (point-wise), in1 = cur (slid)
        const float prev = __ldg(in0 + (g.oz + p.ghost) * p.plane + g.oy * p.row + g.ox);
        const int64_t gz = p.z_off + g.oz;
        if (p.radius == 1) {
          const int K = acoustic_K<1, int64_t>(gz, g.oy, g.ox, p.gnz, p.n[1], p.n[2]);
          v = op_acoustic<1>(CentredAcc{p, in1, g}, prev, K, p.prm);
        } else {
          const int K = acoustic_K<2, int64_t>(gz, g.oy, g.ox, p.gnz, p.n[1], p.n[2]);
          v = op_acoustic<2>(CentredAcc{p, in1, g}, prev, K, p.prm);
        }
        break;
      }
      default:
        v = 0.0f;
    }
    out[(g.oz + p.ghost) * out_plane + g.oy * o2 + g.ox] = v;
  }
}

}  // namespace

cudaError_t launch_generic(const StencilParams& p, const float* in0, const float* in1, float* out,
                           cudaStream_t stream, int num_sms) {
  const int64_t total = (p.reg1 - p.reg0) * p.o[1] * p.o[2];
  if (total <= 0) return cudaSuccess;
  const int threads = 256;
  int64_t blocks = (total + threads - 1) / threads;
  const int64_t cap = (int64_t)num_sms * 8 * 4;   // grid-stride beyond a few waves
  if (blocks > cap) blocks = cap;
  const bool fz = p.put_lo || p.put_hi || p.fused_step || p.wait_lo || p.wait_hi;
  void* args[] = {(void*)&p, (void*)&in0, (void*)&in1, (void*)&out};
  set_last_kernel("k0_generic");
  return launch_kernel(reinterpret_cast<const void*>(&k0_generic), dim3((unsigned)blocks), dim3(threads), args, 0,
                       stream, !fz);
}

}  // namespace lift
