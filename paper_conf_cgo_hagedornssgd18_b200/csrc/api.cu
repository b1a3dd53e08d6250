// api.cu — the C ABI of include/stencil.h: plan creation and validation
// (the pad/slide/map types of PAPER.md P:416-422),
// kernel-family dispatch, apply / apply_region / iterate / run_host.
#include <cuda_runtime.h>

#include <cmath>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <mutex>
#include <new>
#include <string>
#include <utility>
#include <vector>

#include "../../include/stencil.h"
#include "common.cuh"
#include "launch.hpp"
#include "ops.cuh"

using namespace lift;

struct stencil_plan_s {
  int device = 0;
  int ndim = 0;
  int num_sms = 148;
  StencilParams p{};
  int64_t user_out_ext[3] = {0, 0, 0};
  int32_t forced_variant = STENCIL_VARIANT_AUTO;
  int32_t time_block = 0;          // stencil_iterate steps per pass: 0 AUTO (2 where K2R applies), 1, 2
  int32_t last_variant = STENCIL_VARIANT_GENERIC;
  const char* last_kernel = "none";  // kernel function of the most recent launch (stencil_plan_last_kernel)
  // OP_SRAD: device workspace {2 x partials of the q0 reduction, q0 constants}
  void* srad_ws = nullptr;
  // OP_SRAD inside stencil_iterate: the fused pass left the statistics of the
  // image it wrote (srad_chain_img) in partials buffer srad_chain_buf
  // (srad_chain_n entries), so the next pass skips the reduction over I.
  // Only set while stencil_iterate runs (between API calls the caller may
  // rewrite any buffer).
  bool srad_chain = false;
  const float* srad_chain_img = nullptr;
  int srad_chain_buf = 0;
  int srad_chain_n = 0;
  // stencil_run_host workspace (device)
  std::vector<float*> ws;
  size_t ws_elems = 0;
  // stencil_run_host_batch workspace: 3 slots x 4 grids
  std::vector<float*> wsb;
  size_t wsb_elems = 0;
};

namespace {

thread_local std::string g_last_error;

stencil_status fail(stencil_status s, const std::string& msg) {
  g_last_error = msg;
  return s;
}

stencil_status cuda_fail(cudaError_t e, const char* what) {
  g_last_error = std::string(what) + ": " + cudaGetErrorString(e);
  return STENCIL_E_CUDA;
}

// ---- bounded halo waits (fused slab path) --------------------------------
// One process-wide fault block in mapped pinned host memory: a wait that
// times out stores 1 into the word of its code (device store, system scope)
// and the host reads it without a device round trip.  The timeout is
// process-wide too.
std::mutex g_fault_mu;
unsigned int* g_fault = nullptr;          // host pointer == device pointer (UVA)
unsigned long long g_wait_timeout_ns = [] {
  const char* e = getenv("LIFT_WAIT_TIMEOUT_MS");
  return (unsigned long long)(e ? strtoull(e, nullptr, 10) : 10000ull) * 1000000ull;
}();

unsigned int* fault_word(cudaError_t* err) {
  std::lock_guard<std::mutex> lk(g_fault_mu);
  if (!g_fault) {
    void* h = nullptr;
    *err = cudaHostAlloc(&h, 64, cudaHostAllocMapped | cudaHostAllocPortable);
    if (*err != cudaSuccess) return nullptr;
    std::memset(h, 0, 64);
    g_fault = static_cast<unsigned int*>(h);
  }
  *err = cudaSuccess;
  return g_fault;
}

// E_CUDA (and clears the word) if a kernel recorded a fault since the last check
stencil_status take_fault() {
  unsigned int f = 0;
  {
    std::lock_guard<std::mutex> lk(g_fault_mu);
    if (!g_fault) return STENCIL_OK;
    // one word per code (the device stores 1, host memory has no device atomics)
    if (__atomic_exchange_n(&g_fault[kFaultWaitLo - 1], 0u, __ATOMIC_ACQ_REL)) f |= kFaultWaitLo;
    if (__atomic_exchange_n(&g_fault[kFaultWaitHi - 1], 0u, __ATOMIC_ACQ_REL)) f |= kFaultWaitHi;
  }
  if (!f) return STENCIL_OK;
  std::string which = (f & kFaultWaitLo) && (f & kFaultWaitHi) ? "lower and upper"
                      : (f & kFaultWaitLo) ? "lower" : "upper";
  return fail(STENCIL_E_CUDA, "fused halo wait timed out after " + std::to_string(g_wait_timeout_ns / 1000000ull) +
                                  " ms: the " + which +
                                  " neighbour never raised its flag (dead or stalled rank); the step's ghost "
                                  "planes are stale");
}

// Arms a launch's bounded waits.
stencil_status arm_waits(StencilParams& p) {
  cudaError_t e;
  p.fault = fault_word(&e);
  if (!p.fault) return cuda_fail(e, "cudaHostAlloc (fault word)");
  p.wait_timeout_ns = g_wait_timeout_ns;
  return STENCIL_OK;
}

// Saves/restores the caller's current device around library calls.
struct DeviceGuard {
  int prev = -1;
  cudaError_t err = cudaSuccess;
  explicit DeviceGuard(int dev) {
    err = cudaGetDevice(&prev);
    if (err == cudaSuccess && prev != dev) err = cudaSetDevice(dev);
  }
  ~DeviceGuard() {
    int cur = -1;
    if (prev >= 0 && cudaGetDevice(&cur) == cudaSuccess && cur != prev) cudaSetDevice(prev);
  }
};

int op_arity(int op) {
  switch (op) {
    case OP_WEIGHTED: return 1;
    case OP_HOTSPOT3D: return 2;
    case OP_SRAD1: return 1;
    case OP_SRAD2: return 2;
    case OP_ACOUSTIC: return 2;
    case OP_HOTSPOT2D: return 2;
    case OP_GRADIENT: return 1;
    case OP_SRAD: return 1;
    default: return -1;
  }
}

// index of the slid input(s) for aliasing checks: bit i set if input i is slid
int slid_mask(int op) {
  switch (op) {
    case OP_WEIGHTED: return 1;
    case OP_HOTSPOT3D: return 1;      // T slid, P point-wise
    case OP_SRAD1: return 1;
    case OP_SRAD2: return 3;          // c and I both slid
    case OP_ACOUSTIC: return 2;       // prev point-wise, cur slid
    case OP_HOTSPOT2D: return 1;      // T slid, P point-wise
    case OP_GRADIENT: return 1;
    case OP_SRAD: return 1;
    default: return 0;
  }
}

bool same_extents(const StencilParams& p) {
  return p.o[0] == p.n[0] && p.o[1] == p.n[1] && p.o[2] == p.n[2];
}

bool aligned16(const void* ptr) { return (reinterpret_cast<uintptr_t>(ptr) & 15u) == 0; }

int choose_variant(stencil_plan_s* pl, const float* in0, const float* in1, const float* out) {
  const StencilParams& p = pl->p;
  const bool ptr_ok = aligned16(in0) && (in1 == nullptr || aligned16(in1)) && aligned16(out);
  auto want = [&](int v) {
    if (v == STENCIL_VARIANT_SWEEP3D) return ptr_ok && sweep3d_supported(p);
    // K1 fills its tiles with cp.async when TMA cannot (unaligned / nx % 4 != 0)
    if (v == STENCIL_VARIANT_TILE2D) return tile2d_supported(p) && (p.op != OP_SRAD || ptr_ok);
    if (v == STENCIL_VARIANT_GATHER) return gather_supported(p);
    return v == STENCIL_VARIANT_GENERIC;
  };
  if (pl->forced_variant != STENCIL_VARIANT_AUTO)
    return want(pl->forced_variant) ? pl->forced_variant : -1;
  if (pl->ndim == 3 && want(STENCIL_VARIANT_SWEEP3D)) return STENCIL_VARIANT_SWEEP3D;
  if (pl->ndim == 2 && want(STENCIL_VARIANT_TILE2D)) return STENCIL_VARIANT_TILE2D;
  // WEIGHTED plans the TMA families do not take (strided, asymmetric, 1D, wide
  // boxes, unaligned 3D): shared-memory tiles (K5) instead of K0's per-tap loads
  if (want(STENCIL_VARIANT_GATHER)) return STENCIL_VARIANT_GATHER;
  return STENCIL_VARIANT_GENERIC;
}

stencil_status launch(stencil_plan_s* pl, const StencilParams& p_in, const float* in0, const float* in1,
                      float* out, cudaStream_t stream) {
  StencilParams p = p_in;
  const int v = choose_variant(pl, in0, in1, out);
  if (v < 0) return fail(STENCIL_E_UNSUPPORTED, "forced kernel variant cannot run this plan/pointers");
  pl->last_variant = v;
  if (p.op == OP_SRAD) {
    if (!pl->srad_ws) {
      cudaError_t e = cudaMalloc(&pl->srad_ws, srad_workspace_bytes(pl->num_sms));
      if (e != cudaSuccess) return cuda_fail(e, "cudaMalloc (SRAD workspace)");
    }
    const int64_t npts = p.n[1] * p.n[2];
    if (v == STENCIL_VARIANT_TILE2D) {
      // K1S: q0 from partials of in0 (reduced inside the pass), which also
      // writes the partials of out; the image is read for q0 only when no
      // earlier pass of this iterate chain left its statistics
      int src = 0, n_in = 0;
      if (pl->srad_chain && pl->srad_chain_img == in0 && pl->srad_chain_n > 0) {
        src = pl->srad_chain_buf;
        n_in = pl->srad_chain_n;
      } else {
        cudaError_t e = launch_srad_partials(in0, npts, srad_partials_ptr(pl->srad_ws, pl->num_sms, 0), pl->num_sms,
                                             stream, &n_in);
        if (e != cudaSuccess) return cuda_fail(e, "SRAD q0 partials");
      }
      p.srad_part_in = srad_partials_ptr(pl->srad_ws, pl->num_sms, src);
      p.srad_nparts = n_in;
      p.srad_part_out = srad_partials_ptr(pl->srad_ws, pl->num_sms, 1 - src);
      std::string err;
      int n_out = 0;
      cudaError_t e = launch_srad_fused(p, in0, out, stream, pl->num_sms, &err, &n_out);
      pl->last_kernel = g_last_kernel;
      if (e != cudaSuccess)
        return fail(STENCIL_E_CUDA, std::string("kernel launch failed: ") + cudaGetErrorString(e) + " " + err);
      if (pl->srad_chain) {
        pl->srad_chain_img = out;
        pl->srad_chain_buf = 1 - src;
        pl->srad_chain_n = n_out;
      }
      return STENCIL_OK;
    }
    // generic kernel: q0^2 of the current image first (deterministic fp64 reduction)
    cudaError_t e = launch_srad_q0(in0, npts, pl->srad_ws, pl->num_sms, stream);
    if (e != cudaSuccess) return cuda_fail(e, "SRAD q0 reduction");
    p.srad_q0 = srad_q0_ptr(pl->srad_ws, pl->num_sms);
  }
  std::string err;
  cudaError_t e;
  set_last_kernel("none");
  switch (v) {
    case STENCIL_VARIANT_SWEEP3D:
      e = launch_sweep3d(p, in0, in1, out, stream, pl->num_sms, &err);
      break;
    case STENCIL_VARIANT_GATHER:
      e = launch_gather(p, in0, out, stream, pl->num_sms, &err);
      break;
    case STENCIL_VARIANT_TILE2D:
      e = launch_tile2d(p, in0, in1, out, stream, pl->num_sms, &err);
      break;
    default:
      e = launch_generic(p, in0, in1, out, stream, pl->num_sms);
  }
  pl->last_kernel = g_last_kernel;
  if (e != cudaSuccess) {
    g_last_error = std::string("kernel launch failed: ") + cudaGetErrorString(e) + (err.empty() ? "" : " (" + err + ")");
    return STENCIL_E_CUDA;
  }
  if (!err.empty()) return fail(STENCIL_E_CUDA, err);
  return STENCIL_OK;
}

stencil_status check_inputs(stencil_plan_s* pl, const float* const* inputs, int32_t n_inputs,
                            const float* out) {
  const int ar = op_arity(pl->p.op);
  if (n_inputs != ar) return fail(STENCIL_E_INVALID, "n_inputs does not match the op's arity");
  if (!inputs || !out) return fail(STENCIL_E_INVALID, "NULL input/output pointer");
  for (int i = 0; i < n_inputs; ++i)
    if (!inputs[i]) return fail(STENCIL_E_INVALID, "NULL input pointer");
  const int m = slid_mask(pl->p.op);
  for (int i = 0; i < n_inputs; ++i)
    if ((m >> i) & 1)
      if (inputs[i] == out) return fail(STENCIL_E_INVALID, "output aliases a slid input");
  return STENCIL_OK;
}

}  // namespace

extern "C" {

const char* stencil_version(void) { return "lift-stencil-b200 0.1 (sm_100a)"; }

const char* stencil_status_string(stencil_status s) {
  switch (s) {
    case STENCIL_OK: return "ok";
    case STENCIL_E_INVALID: return "invalid argument";
    case STENCIL_E_UNSUPPORTED: return "unsupported";
    case STENCIL_E_CUDA: return "CUDA error";
    case STENCIL_E_NOMEM: return "out of memory";
  }
  return "unknown status";
}

const char* stencil_last_error(void) { return g_last_error.c_str(); }

stencil_status stencil_plan_create(stencil_plan* out, int device, int ndim, const int64_t* extents,
                                   const int32_t* size, const int32_t* step, const int32_t* pad_lo,
                                   const int32_t* pad_hi, const int32_t* kind, float pad_value,
                                   int32_t op, const float* weights, const float* params,
                                   int32_t n_params) {
  if (!out) return fail(STENCIL_E_INVALID, "out is NULL");
  *out = nullptr;
  if (ndim > 3) return fail(STENCIL_E_UNSUPPORTED, "ndim > 3 is not built");
  if (ndim < 1) return fail(STENCIL_E_INVALID, "ndim must be 1, 2 or 3");
  if (!extents || !size || !step || !pad_lo || !pad_hi || !kind)
    return fail(STENCIL_E_INVALID, "NULL array argument");
  if (op < 0 || op > OP_SRAD) return fail(STENCIL_E_INVALID, "unknown op");
  if (n_params < 0 || n_params > kMaxParams || (n_params > 0 && !params))
    return fail(STENCIL_E_INVALID, "bad params");

  StencilParams p{};
  const int off = 3 - ndim;
  for (int d = 0; d < 3; ++d) {
    p.n[d] = 1; p.size[d] = 1; p.step[d] = 1; p.lo[d] = 0; p.hi[d] = 0; p.kind[d] = PAD_CLAMP;
  }
  for (int d = 0; d < ndim; ++d) {
    if (extents[d] < 1 || size[d] < 1 || step[d] < 1 || pad_lo[d] < 0 || pad_hi[d] < 0)
      return fail(STENCIL_E_INVALID, "extents/size/step must be >= 1 and pads >= 0");
    if (kind[d] < PAD_CLAMP || kind[d] > PAD_DAMPEN) return fail(STENCIL_E_INVALID, "unknown pad kind");
    if (kind[d] == PAD_DAMPEN && op != OP_WEIGHTED)
      return fail(STENCIL_E_UNSUPPORTED, "DAMPEN pads are built for WEIGHTED stencils");
    if (extents[d] + pad_lo[d] + pad_hi[d] < size[d])
      return fail(STENCIL_E_INVALID, "n + l + r < size: slide yields no window");
    if (extents[d] > (int64_t)1 << 40 || size[d] > 4096 || pad_lo[d] > (1 << 20) || pad_hi[d] > (1 << 20))
      return fail(STENCIL_E_INVALID, "extent/size/pad out of supported range");
    p.n[off + d] = extents[d];
    p.size[off + d] = size[d];
    p.step[off + d] = step[d];
    p.lo[off + d] = pad_lo[d];
    p.hi[off + d] = pad_hi[d];
    p.kind[off + d] = kind[d];
  }
  for (int d = 0; d < 3; ++d) p.o[d] = (p.n[d] + p.lo[d] + p.hi[d] - p.size[d]) / p.step[d] + 1;
  p.row = p.n[2];
  p.plane = p.n[1] * p.n[2];
  p.pad_value = pad_value;
  p.pad_decay = 1.0f;
  p.op = op;
  p.z_off = 0;
  p.gnz = p.n[0];
  p.ghost = 0;
  p.slab = 0;
  p.reg0 = 0;
  p.reg1 = p.o[0];
  for (int i = 0; i < n_params; ++i) p.prm[i] = params[i];

  // op-specific shape rules (stencil.h / DESIGN.md A16-A20)
  auto centred = [&](int r) {
    for (int d = off; d < 3; ++d)
      if (p.size[d] != 2 * r + 1 || p.lo[d] != r || p.hi[d] != r || p.step[d] != 1) return false;
    return true;
  };
  switch (op) {
    case OP_WEIGHTED: {
      if (!weights) return fail(STENCIL_E_INVALID, "WEIGHTED needs weights");
      int64_t ntot = 1;
      for (int d = 0; d < ndim; ++d) ntot *= size[d];
      if (ntot > (int64_t)1 << 24) return fail(STENCIL_E_INVALID, "window too large");
      int nt = 0;
      const int64_t s1 = p.size[1], s2 = p.size[2];
      for (int64_t k = 0; k < ntot; ++k) {
        if (weights[k] == 0.0f) continue;
        if (nt >= kMaxTaps) return fail(STENCIL_E_UNSUPPORTED, "more than 125 non-zero taps");
        const int64_t kz = k / (s1 * s2), ky = (k / s2) % s1, kx = k % s2;
        p.tap[nt][0] = (int16_t)kz;
        p.tap[nt][1] = (int16_t)ky;
        p.tap[nt][2] = (int16_t)kx;
        p.w[nt] = weights[k];
        ++nt;
      }
      p.ntaps = nt;
      {
        // linear tap offsets for K0's interior fast path (needs 32-bit offsets)
        const int64_t span = (int64_t)(p.size[0] - 1) * p.plane + (int64_t)(p.size[1] - 1) * p.row + p.size[2];
        if (span < ((int64_t)1 << 31))
          for (int t = 0; t < nt; ++t)
            p.tap_off[t] = (int32_t)(p.tap[t][0] * p.plane + p.tap[t][1] * p.row + p.tap[t][2]);
        else if (nt > 0)
          p.tap_off[0] = -1;
      }
      if (ntot <= kMaxTaps)
        for (int64_t k = 0; k < ntot; ++k) p.wbox[k] = weights[k];
      // separable (rank-1) 2D weights: w[i][j] == su[i] * sv[j] exactly (checked
      // in double, where fp32 x fp32 products are exact); the factors are scaled
      // by sqrt of the largest tap so that e.g. the binomial Gaussian factors
      // into its exact 1D binomials
      p.sep = 0;
      if (ndim == 2 && p.size[1] <= kMaxSep && p.size[2] <= kMaxSep) {
        const int SY = p.size[1], SX = p.size[2];
        int bi = 0, bj = 0;
        for (int i = 0; i < SY; ++i)
          for (int j = 0; j < SX; ++j)
            if (std::fabs(weights[i * SX + j]) > std::fabs(weights[bi * SX + bj])) { bi = i; bj = j; }
        const float wc = weights[bi * SX + bj];
        if (wc != 0.0f) {
          const float sc = std::sqrt(std::fabs(wc));
          float u[kMaxSep], v[kMaxSep];
          for (int j = 0; j < SX; ++j) v[j] = weights[bi * SX + j] / sc;
          for (int i = 0; i < SY; ++i) u[i] = weights[i * SX + bj] / (wc / sc);
          bool ok = true;
          for (int i = 0; i < SY && ok; ++i)
            for (int j = 0; j < SX && ok; ++j)
              ok = (double)u[i] * (double)v[j] == (double)weights[i * SX + j];
          if (ok) {
            p.sep = 1;
            for (int i = 0; i < SY; ++i) p.su[i] = u[i];
            for (int j = 0; j < SX; ++j) p.sv[j] = v[j];
          }
        }
      }
      // radius for the fast kernels: symmetric centred window
      int r = p.size[2] / 2;
      p.radius = centred(r) ? r : -1;
      break;
    }
    case OP_HOTSPOT3D:
      if (ndim != 3 || !centred(1)) return fail(STENCIL_E_INVALID, "HOTSPOT3D needs ndim 3, size 3, pad 1, step 1");
      if (n_params < 9) return fail(STENCIL_E_INVALID, "HOTSPOT3D needs 9 params");
      p.radius = 1;
      break;
    case OP_SRAD1:
    case OP_SRAD2:
      if (ndim != 2 || !centred(1)) return fail(STENCIL_E_INVALID, "SRAD needs ndim 2, size 3, pad 1, step 1");
      if (n_params < 1) return fail(STENCIL_E_INVALID, "SRAD needs 1 param");
      if (op == OP_SRAD1) {
        if (!(params[0] > 0.0f)) return fail(STENCIL_E_INVALID, "SRAD1 needs q0sqr > 0");
        srad1_constants(params[0], p.prm);                // derived plan constants (A18b)
      }
      p.radius = 1;
      break;
    case OP_HOTSPOT2D:
      if (ndim != 2 || !centred(1)) return fail(STENCIL_E_INVALID, "HOTSPOT2D needs ndim 2, size 3, pad 1, step 1");
      if (n_params < 5) return fail(STENCIL_E_INVALID, "HOTSPOT2D needs 5 params");
      p.radius = 1;
      break;
    case OP_SRAD:
      if (ndim != 2 || !centred(1)) return fail(STENCIL_E_INVALID, "SRAD needs ndim 2, size 3, pad 1, step 1");
      if (n_params < 1) return fail(STENCIL_E_INVALID, "SRAD needs 1 param (lambda)");
      if (kind[0] == PAD_CONSTANT || kind[1] == PAD_CONSTANT)
        return fail(STENCIL_E_UNSUPPORTED, "SRAD iteration is built for reindexing pads");
      p.radius = 1;
      break;
    case OP_GRADIENT:
      if (ndim != 2 || !centred(1)) return fail(STENCIL_E_INVALID, "GRADIENT needs ndim 2, size 3, pad 1, step 1");
      if (n_params < 1) return fail(STENCIL_E_INVALID, "GRADIENT needs 1 param (eps)");
      p.radius = 1;
      break;
    case OP_ACOUSTIC:
      if (ndim != 3 || !(centred(1) || centred(2)))
        return fail(STENCIL_E_INVALID, "ACOUSTIC needs ndim 3, size 3 or 5, pad r, step 1");
      if (n_params < 3) return fail(STENCIL_E_INVALID, "ACOUSTIC needs 3 params");
      p.radius = p.size[2] / 2;
      break;
  }

  stencil_plan_s* pl = new (std::nothrow) stencil_plan_s();
  if (!pl) return fail(STENCIL_E_NOMEM, "plan allocation failed");
  pl->device = device;
  pl->ndim = ndim;
  pl->p = p;
  for (int d = 0; d < ndim; ++d) pl->user_out_ext[d] = p.o[off + d];
  int sms = 0;
  if (cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, device) == cudaSuccess && sms > 0)
    pl->num_sms = sms;
  else
    cudaGetLastError();  // no device here: plan creation is host-only
  *out = pl;
  return STENCIL_OK;
}

stencil_status stencil_plan_output_extents(stencil_plan pl, int64_t* out_ext) {
  if (!pl || !out_ext) return fail(STENCIL_E_INVALID, "NULL argument");
  for (int d = 0; d < pl->ndim; ++d) out_ext[d] = pl->user_out_ext[d];
  return STENCIL_OK;
}

stencil_status stencil_plan_set_slab(stencil_plan pl, int64_t z_offset, int64_t global_n0, int32_t ghost) {
  if (!pl) return fail(STENCIL_E_INVALID, "NULL plan");
  StencilParams& p = pl->p;
  if (pl->ndim != 3) return fail(STENCIL_E_UNSUPPORTED, "slab mode is built for 3D plans");
  if (!same_extents(p) || p.step[0] != 1) return fail(STENCIL_E_INVALID, "slab mode needs output extents == input extents and step 1");
  if (ghost < p.lo[0] || ghost < p.hi[0]) return fail(STENCIL_E_INVALID, "ghost < pad in dimension 0");
  if (z_offset < 0 || global_n0 < z_offset + p.n[0]) return fail(STENCIL_E_INVALID, "slab outside the global grid");
  p.z_off = z_offset;
  p.gnz = global_n0;
  p.ghost = ghost;
  p.slab = 1;
  // allocate the fault word now, outside any graph capture (without a device
  // this fails quietly; the fused launches retry and report it)
  cudaError_t e;
  (void)fault_word(&e);
  return STENCIL_OK;
}

stencil_status stencil_plan_set_variant(stencil_plan pl, int32_t variant) {
  if (!pl) return fail(STENCIL_E_INVALID, "NULL plan");
  if (variant < STENCIL_VARIANT_AUTO || variant > STENCIL_VARIANT_GATHER || variant == STENCIL_VARIANT_PERSIST3D)
    return fail(STENCIL_E_INVALID, "unknown or non-forceable variant");
  if (variant == STENCIL_VARIANT_GATHER && !gather_supported(pl->p))
    return fail(STENCIL_E_UNSUPPORTED, "GATHER cannot run this plan");
  if (variant == STENCIL_VARIANT_SWEEP3D && !sweep3d_supported(pl->p))
    return fail(STENCIL_E_UNSUPPORTED, "SWEEP3D cannot run this plan");
  if (variant == STENCIL_VARIANT_TILE2D && !tile2d_supported(pl->p))
    return fail(STENCIL_E_UNSUPPORTED, "TILE2D cannot run this plan");
  pl->forced_variant = variant;
  return STENCIL_OK;
}

stencil_status stencil_plan_set_time_block(stencil_plan pl, int32_t steps) {
  if (!pl) return fail(STENCIL_E_INVALID, "NULL plan");
  if (steps < 0 || steps > 2) return fail(STENCIL_E_INVALID, "time block must be 0 (auto), 1 or 2");
  pl->time_block = steps;
  return STENCIL_OK;
}

int32_t stencil_plan_time_block(stencil_plan pl) {
  if (!pl) return -1;
  const bool hs2 = pl->p.op == OP_HOTSPOT3D && column3d_t2_supported(pl->p, nullptr, nullptr);
  // (K2CT, two Hotspot3D steps per launch of a few-plane grid, measured no
  // faster than K2C single steps — 6.75 vs 6.53 us per step — so AUTO keeps
  // single steps for it; time block 2 forces it)
  if (pl->time_block == 0)
    return (pl->ndim == 3 && (sweep3d_r2_auto(pl->p) || acoustic_r2_auto(pl->p))) ? 2 : 1;
  return (pl->time_block >= 2 && pl->ndim == 3 &&
          (sweep3d_t2_supported(pl->p) || acoustic_r2_supported(pl->p) || hs2))
             ? 2
             : 1;
}

int32_t stencil_plan_last_variant(stencil_plan pl) { return pl ? pl->last_variant : -1; }

const char* stencil_plan_last_kernel(stencil_plan pl) { return pl ? pl->last_kernel : "none"; }

stencil_status stencil_plan_set_pad_decay(stencil_plan pl, float decay) {
  if (!pl) return fail(STENCIL_E_INVALID, "NULL plan");
  if (!(decay >= 0.0f && decay <= 1.0f)) return fail(STENCIL_E_INVALID, "pad decay must be in [0, 1]");
  pl->p.pad_decay = decay;
  return STENCIL_OK;
}

int32_t stencil_plan_variant(stencil_plan pl) {
  if (!pl) return -1;
  if (pl->forced_variant != STENCIL_VARIANT_AUTO) return pl->forced_variant;
  const StencilParams& p = pl->p;
  if (pl->ndim == 3 && sweep3d_supported(p)) return STENCIL_VARIANT_SWEEP3D;
  if (pl->ndim == 2 && tile2d_supported(p)) return STENCIL_VARIANT_TILE2D;
  if (gather_supported(p)) return STENCIL_VARIANT_GATHER;
  return STENCIL_VARIANT_GENERIC;
}

stencil_status stencil_apply_region(stencil_plan pl, const float* const* inputs, int32_t n_inputs,
                                    float* out, int64_t o0_begin, int64_t o0_end, void* stream) {
  if (!pl) return fail(STENCIL_E_INVALID, "NULL plan");
  stencil_status s = check_inputs(pl, inputs, n_inputs, out);
  if (s != STENCIL_OK) return s;
  // region is along the plan's dimension 0 (the slowest user dimension)
  const int off = 3 - pl->ndim;
  if (off != 0) {
    if (!(o0_begin == 0 && o0_end == pl->user_out_ext[0]))
      return fail(STENCIL_E_UNSUPPORTED, "apply_region is built for 3D plans");
    o0_begin = 0;            // canonical dimension 0 has extent 1
    o0_end = pl->p.o[0];
  }
  // slab plans may extend the region into the ghost planes (deep halos,
  // NEXT-3: the overlap of k time steps is recomputed redundantly) as far as
  // the window's input planes stay inside the allocation
  int64_t lo_lim = 0, hi_lim = pl->p.o[0];
  if (pl->p.slab) {
    lo_lim = -(int64_t)(pl->p.ghost - pl->p.lo[0]);
    hi_lim = pl->p.o[0] + (pl->p.ghost - pl->p.hi[0]);
  }
  if (o0_begin < lo_lim || o0_end > hi_lim || o0_begin > o0_end)
    return fail(STENCIL_E_INVALID, "region outside the output extents (slab: ghost planes minus the pad)");
  if (o0_begin == o0_end) return STENCIL_OK;
  DeviceGuard g(pl->device);
  if (g.err != cudaSuccess) return cuda_fail(g.err, "cudaSetDevice");
  StencilParams p = pl->p;
  p.reg0 = o0_begin;
  p.reg1 = o0_end;
  return launch(pl, p, inputs[0], n_inputs > 1 ? inputs[1] : nullptr, out, (cudaStream_t)stream);
}

stencil_status stencil_apply2_region(stencil_plan pl, const float* in, float* out, int64_t o0_begin, int64_t o0_end,
                                     void* stream) {
  if (!pl) return fail(STENCIL_E_INVALID, "NULL plan");
  if (!in || !out || in == out) return fail(STENCIL_E_INVALID, "apply2_region: bad or aliasing buffers");
  if (pl->ndim != 3 || !sweep3d_t2_supported(pl->p))
    return fail(STENCIL_E_UNSUPPORTED, "apply2_region: no two-step kernel takes this plan");
  if (!aligned16(in) || !aligned16(out)) return fail(STENCIL_E_INVALID, "apply2_region: buffers must be 16-B aligned");
  int64_t lo_lim = 0, hi_lim = pl->p.o[0];
  if (pl->p.slab) {
    lo_lim = -(int64_t)(pl->p.ghost - 2 * pl->p.lo[0]);
    hi_lim = pl->p.o[0] + (pl->p.ghost - 2 * pl->p.hi[0]);
  }
  if (o0_begin < lo_lim || o0_end > hi_lim || o0_begin > o0_end)
    return fail(STENCIL_E_INVALID, "apply2_region: region outside the output extents (slab: ghosts minus 2 pads)");
  if (o0_begin == o0_end) return STENCIL_OK;
  DeviceGuard g(pl->device);
  if (g.err != cudaSuccess) return cuda_fail(g.err, "cudaSetDevice");
  StencilParams p = pl->p;
  p.reg0 = o0_begin;
  p.reg1 = o0_end;
  std::string err;
  cudaError_t e = launch_sweep3d_t2(p, in, out, (cudaStream_t)stream, pl->num_sms, &err);
  pl->last_kernel = g_last_kernel;
  pl->last_variant = STENCIL_VARIANT_SWEEP3D;
  if (e != cudaSuccess) return fail(STENCIL_E_CUDA, std::string("two-step launch failed: ") + cudaGetErrorString(e) + " " + err);
  return STENCIL_OK;
}

stencil_status stencil_apply_region_put(stencil_plan pl, const float* const* inputs, int32_t n_inputs, float* out,
                                        int64_t o0_begin, int64_t o0_end, float* put_lo, float* put_hi,
                                        uint32_t* sig_lo, uint32_t* sig_hi, uint32_t sig_value, void* stream) {
  if (!pl) return fail(STENCIL_E_INVALID, "NULL plan");
  stencil_status s = check_inputs(pl, inputs, n_inputs, out);
  if (s != STENCIL_OK) return s;
  if (!pl->p.slab) return fail(STENCIL_E_INVALID, "fused halo put needs a slab plan (stencil_plan_set_slab)");
  s = take_fault();
  if (s != STENCIL_OK) return s;
  if (o0_begin < 0 || o0_end > pl->p.o[0] || o0_begin >= o0_end)
    return fail(STENCIL_E_INVALID, "region outside the output extents");
  if (choose_variant(pl, inputs[0], n_inputs > 1 ? inputs[1] : nullptr, out) != STENCIL_VARIANT_SWEEP3D)
    return fail(STENCIL_E_UNSUPPORTED, "fused halo put is built on the TMA sweep kernel only");
  DeviceGuard g(pl->device);
  if (g.err != cudaSuccess) return cuda_fail(g.err, "cudaSetDevice");
  StencilParams p = pl->p;
  p.reg0 = o0_begin;
  p.reg1 = o0_end;
  p.put_lo = put_lo;
  p.put_hi = put_hi;
  p.sig_lo = sig_lo;
  p.sig_hi = sig_hi;
  p.sig_value = sig_value;
  return launch(pl, p, inputs[0], n_inputs > 1 ? inputs[1] : nullptr, out, (cudaStream_t)stream);
}

stencil_status stencil_slab_step_fused(stencil_plan pl, const float* const* inputs, int32_t n_inputs, float* out,
                                       float* put_lo, float* put_hi, uint32_t* sig_lo, uint32_t* sig_hi,
                                       uint32_t sig_value, const uint32_t* wait_lo, const uint32_t* wait_hi,
                                       uint32_t wait_value, void* stream) {
  if (!pl) return fail(STENCIL_E_INVALID, "NULL plan");
  stencil_status s = check_inputs(pl, inputs, n_inputs, out);
  if (s != STENCIL_OK) return s;
  if (!pl->p.slab) return fail(STENCIL_E_INVALID, "fused step needs a slab plan (stencil_plan_set_slab)");
  s = take_fault();
  if (s != STENCIL_OK) return s;
  if (choose_variant(pl, inputs[0], n_inputs > 1 ? inputs[1] : nullptr, out) != STENCIL_VARIANT_SWEEP3D)
    return fail(STENCIL_E_UNSUPPORTED, "fused step is built on the TMA sweep kernel only");
  DeviceGuard g(pl->device);
  if (g.err != cudaSuccess) return cuda_fail(g.err, "cudaSetDevice");
  StencilParams p = pl->p;
  p.reg0 = 0;
  p.reg1 = p.o[0];
  p.put_lo = put_lo;
  p.put_hi = put_hi;
  p.sig_lo = sig_lo;
  p.sig_hi = sig_hi;
  p.sig_value = sig_value;
  p.wait_lo = wait_lo;
  p.wait_hi = wait_hi;
  p.wait_value = wait_value;
  p.fused_step = 1;
  s = arm_waits(p);
  if (s != STENCIL_OK) return s;
  return launch(pl, p, inputs[0], n_inputs > 1 ? inputs[1] : nullptr, out, (cudaStream_t)stream);
}

stencil_status stencil_wait_signals(const uint32_t* sig_a, const uint32_t* sig_b, uint32_t value, void* stream) {
  stencil_status s = take_fault();
  if (s != STENCIL_OK) return s;
  cudaError_t e;
  unsigned int* fault = fault_word(&e);
  if (!fault) return cuda_fail(e, "cudaHostAlloc (fault word)");
  e = launch_wait_signals(sig_a, sig_b, value, g_wait_timeout_ns, fault, (cudaStream_t)stream);
  if (e != cudaSuccess) return cuda_fail(e, "wait kernel launch");
  return STENCIL_OK;
}

stencil_status stencil_set_wait_timeout_ms(uint32_t ms) {
  std::lock_guard<std::mutex> lk(g_fault_mu);
  g_wait_timeout_ns = (unsigned long long)ms * 1000000ull;
  return STENCIL_OK;
}

stencil_status stencil_device_fault(void) { return take_fault(); }

stencil_status stencil_apply(stencil_plan pl, const float* const* inputs, int32_t n_inputs, float* out,
                             void* stream) {
  if (!pl) return fail(STENCIL_E_INVALID, "NULL plan");
  return stencil_apply_region(pl, inputs, n_inputs, out, 0, pl->user_out_ext[0], stream);
}

stencil_status stencil_iterate(stencil_plan pl, float* const* state, int32_t n_state, const float* const* aux,
                               int32_t n_aux, int32_t n_steps, void* stream, int32_t* result_index) {
  if (!pl) return fail(STENCIL_E_INVALID, "NULL plan");
  const StencilParams& p = pl->p;
  if (!same_extents(p)) return fail(STENCIL_E_INVALID, "iterate needs output extents == input extents");
  if (n_steps < 0) return fail(STENCIL_E_INVALID, "n_steps < 0");
  if (!state || !(n_state == 2 || (n_state == 4 && p.op == OP_ACOUSTIC)))
    return fail(STENCIL_E_INVALID, "iterate needs 2 state buffers (ACOUSTIC: 2 or 4)");
  for (int i = 0; i < n_state; ++i) {
    if (!state[i]) return fail(STENCIL_E_INVALID, "bad state buffers");
    for (int k = 0; k < i; ++k)
      if (state[k] == state[i]) return fail(STENCIL_E_INVALID, "bad state buffers");
  }
  int ri = (p.op == OP_ACOUSTIC) ? 1 : 0;
  const int32_t tb = stencil_plan_time_block(pl);     // steps per pass (K2R / K2T when 2)
  // few-plane 3D grids that fit in the device's shared memory: all steps in
  // one cooperative launch with the grid resident on chip (K6)
  if ((p.op == OP_WEIGHTED || p.op == OP_HOTSPOT3D) && n_steps >= 2 && pl->ndim == 3 && pl->time_block != 2 &&
      pl->forced_variant == STENCIL_VARIANT_AUTO &&
      (p.op == OP_WEIGHTED ? n_aux == 0 : (n_aux == 1 && aux && aux[0])) &&
      resident3d_supported(p, state[0], state[1], p.op == OP_HOTSPOT3D ? aux[0] : nullptr, pl->num_sms)) {
    DeviceGuard g(pl->device);
    if (g.err != cudaSuccess) return cuda_fail(g.err, "cudaSetDevice");
    std::string err;
    cudaError_t e = launch_resident3d(p, state[0], state[1], p.op == OP_HOTSPOT3D ? aux[0] : nullptr, n_steps,
                                      (cudaStream_t)stream, pl->num_sms, &err);
    if (e != cudaSuccess)
      return fail(STENCIL_E_CUDA, std::string("K6 launch failed: ") + cudaGetErrorString(e) + " " + err);
    pl->last_variant = STENCIL_VARIANT_RESIDENT3D;
    pl->last_kernel = g_last_kernel;
    if (result_index) *result_index = n_steps % 2;
    return STENCIL_OK;
  }
  // small L2-resident 3D grids: all steps in one persistent launch (K4)
  if ((p.op == OP_WEIGHTED || p.op == OP_HOTSPOT3D) && n_steps >= 2 && pl->ndim == 3 && pl->time_block != 2 &&
      pl->forced_variant == STENCIL_VARIANT_AUTO &&
      (p.op == OP_WEIGHTED ? n_aux == 0 : (n_aux == 1 && aux && aux[0])) &&
      persist3d_supported(p, state[0], state[1], p.op == OP_HOTSPOT3D ? aux[0] : nullptr)) {
    DeviceGuard g(pl->device);
    if (g.err != cudaSuccess) return cuda_fail(g.err, "cudaSetDevice");
    std::string err;
    cudaError_t e = launch_persist3d(p, state[0], state[1], p.op == OP_HOTSPOT3D ? aux[0] : nullptr, n_steps,
                                     (cudaStream_t)stream, pl->num_sms, &err);
    if (e != cudaSuccess)
      return fail(STENCIL_E_CUDA, std::string("K4 launch failed: ") + cudaGetErrorString(e) + " " + err);
    pl->last_variant = STENCIL_VARIANT_PERSIST3D;
    pl->last_kernel = g_last_kernel;
    if (result_index) *result_index = n_steps % 2;
    return STENCIL_OK;
  }
  if (p.op == OP_WEIGHTED || p.op == OP_GRADIENT || p.op == OP_SRAD) {
    if (n_aux != 0) return fail(STENCIL_E_INVALID, "WEIGHTED/GRADIENT/SRAD iterate takes no aux grids");
    int t = 0;
    // temporal blocking: two steps per pass (K2T) while at least two remain
    if (tb >= 2 && n_steps >= 2 &&
        (pl->forced_variant == STENCIL_VARIANT_AUTO || pl->forced_variant == STENCIL_VARIANT_SWEEP3D) &&
        aligned16(state[0]) && aligned16(state[1])) {
      DeviceGuard g(pl->device);
      if (g.err != cudaSuccess) return cuda_fail(g.err, "cudaSetDevice");
      for (; t + 2 <= n_steps; t += 2) {
        std::string err;
        cudaError_t e = launch_sweep3d_t2(p, state[ri], state[1 - ri], (cudaStream_t)stream, pl->num_sms, &err);
        pl->last_kernel = g_last_kernel;
        pl->last_variant = STENCIL_VARIANT_SWEEP3D;
        if (e != cudaSuccess)
          return fail(STENCIL_E_CUDA, std::string("K2T launch failed: ") + cudaGetErrorString(e) + " " + err);
        ri = 1 - ri;
      }
    }
    // SRAD: each fused pass hands the statistics of its output to the next
    struct ChainGuard {
      stencil_plan_s* pl;
      ~ChainGuard() {
        pl->srad_chain = false;
        pl->srad_chain_img = nullptr;
        pl->srad_chain_n = 0;
      }
    } chain_guard{pl};
    pl->srad_chain = p.op == OP_SRAD;
    pl->srad_chain_img = nullptr;
    pl->srad_chain_n = 0;
    for (; t < n_steps; ++t) {
      const float* in[1] = {state[ri]};
      stencil_status s = stencil_apply(pl, in, 1, state[1 - ri], stream);
      if (s != STENCIL_OK) return s;
      ri = 1 - ri;
    }
  } else if (p.op == OP_HOTSPOT3D || p.op == OP_HOTSPOT2D) {
    if (n_aux != 1 || !aux || !aux[0]) return fail(STENCIL_E_INVALID, "HOTSPOT iterate needs aux {P}");
    int t = 0;
    // two steps per launch (K2CT) for few-plane Hotspot3D grids
    if (p.op == OP_HOTSPOT3D && tb == 2 && n_steps >= 2 && pl->ndim == 3 &&
        (pl->forced_variant == STENCIL_VARIANT_AUTO || pl->forced_variant == STENCIL_VARIANT_SWEEP3D) &&
        column3d_t2_supported(p, state[0], aux[0]) && column3d_t2_supported(p, state[1], aux[0])) {
      DeviceGuard g(pl->device);
      if (g.err != cudaSuccess) return cuda_fail(g.err, "cudaSetDevice");
      for (; t + 2 <= n_steps; t += 2) {
        std::string err;
        cudaError_t e = launch_column3d_t2(p, state[ri], aux[0], state[1 - ri], (cudaStream_t)stream, &err);
        pl->last_kernel = g_last_kernel;
        pl->last_variant = STENCIL_VARIANT_SWEEP3D;
        if (e != cudaSuccess)
          return fail(STENCIL_E_CUDA, std::string("K2CT launch failed: ") + cudaGetErrorString(e) + " " + err);
        ri = 1 - ri;
      }
    }
    for (; t < n_steps; ++t) {
      const float* in[2] = {state[ri], aux[0]};
      stencil_status s = stencil_apply(pl, in, 2, state[1 - ri], stream);
      if (s != STENCIL_OK) return s;
      ri = 1 - ri;
    }
  } else if (p.op == OP_ACOUSTIC) {
    if (n_aux != 0) return fail(STENCIL_E_INVALID, "ACOUSTIC iterate takes no aux grids");
    // state {prev, cur} (+ two spare grids): (a, b) = (prev, cur)
    int a = 0, b = 1, t = 0;
    if (n_state == 4 && tb == 2 && n_steps >= 2 && pl->ndim == 3 && acoustic_r2_supported(p) &&
        (pl->forced_variant == STENCIL_VARIANT_AUTO || pl->forced_variant == STENCIL_VARIANT_SWEEP3D) &&
        aligned16(state[0]) && aligned16(state[1]) && aligned16(state[2]) && aligned16(state[3])) {
      // K2RA: two steps per pass, (prev, cur) -> (u^{n+1}, u^{n+2}) in the spare pair
      DeviceGuard g(pl->device);
      if (g.err != cudaSuccess) return cuda_fail(g.err, "cudaSetDevice");
      int c = 2, d = 3;
      for (; t + 2 <= n_steps; t += 2) {
        std::string err;
        cudaError_t e = launch_acoustic_r2(p, state[a], state[b], state[c], state[d], (cudaStream_t)stream,
                                           pl->num_sms, &err);
        pl->last_kernel = g_last_kernel;
        pl->last_variant = STENCIL_VARIANT_SWEEP3D;
        if (e != cudaSuccess)
          return fail(STENCIL_E_CUDA, std::string("K2RA launch failed: ") + cudaGetErrorString(e) + " " + err);
        std::swap(a, c);
        std::swap(b, d);
      }
    }
    // single steps: next overwrites prev, then roles swap (A21)
    for (; t < n_steps; ++t) {
      const float* in[2] = {state[a], state[b]};
      stencil_status s = stencil_apply(pl, in, 2, state[a], stream);
      if (s != STENCIL_OK) return s;
      std::swap(a, b);
    }
    ri = b;
  } else {
    return fail(STENCIL_E_UNSUPPORTED, "iterate is built for WEIGHTED, HOTSPOT3D/2D, GRADIENT and ACOUSTIC");
  }
  if (result_index) *result_index = ri;
  return STENCIL_OK;
}

stencil_status stencil_run_host(stencil_plan pl, const float* const* host_state, int32_t n_state,
                                const float* const* host_aux, int32_t n_aux, int32_t n_steps,
                                float* host_out, void* stream) {
  if (!pl) return fail(STENCIL_E_INVALID, "NULL plan");
  if (!host_state || !host_out || n_state < 1 || n_state > 2 || n_aux < 0 || n_aux > 1)
    return fail(STENCIL_E_INVALID, "bad host buffers");
  const StencilParams& p = pl->p;
  DeviceGuard g(pl->device);
  if (g.err != cudaSuccess) return cuda_fail(g.err, "cudaSetDevice");
  cudaStream_t st = (cudaStream_t)stream;
  const size_t in_elems = (size_t)(p.n[0] + 2 * p.ghost) * p.plane;
  const size_t out_elems = (size_t)(p.o[0] + 2 * p.ghost) * p.o[1] * p.o[2];
  const size_t elems = in_elems > out_elems ? in_elems : out_elems;
  const int nbuf = 4;  // state0, state1, aux0, out
  if (pl->ws_elems < elems) {
    for (float* b : pl->ws) cudaFree(b);
    pl->ws.clear();
    pl->ws_elems = 0;
    for (int i = 0; i < nbuf; ++i) {
      float* b = nullptr;
      cudaError_t e = cudaMalloc(&b, elems * sizeof(float));
      if (e != cudaSuccess) return cuda_fail(e, "cudaMalloc (run_host workspace)");
      pl->ws.push_back(b);
    }
    pl->ws_elems = elems;
  }
  cudaError_t e;
  for (int i = 0; i < n_state; ++i) {
    e = cudaMemcpyAsync(pl->ws[i], host_state[i], in_elems * sizeof(float), cudaMemcpyHostToDevice, st);
    if (e != cudaSuccess) return cuda_fail(e, "H2D copy");
  }
  for (int i = 0; i < n_aux; ++i) {
    e = cudaMemcpyAsync(pl->ws[2], host_aux[i], in_elems * sizeof(float), cudaMemcpyHostToDevice, st);
    if (e != cudaSuccess) return cuda_fail(e, "H2D copy");
  }
  const float* result = nullptr;
  const bool iterable = (p.op == OP_WEIGHTED || p.op == OP_HOTSPOT3D || p.op == OP_ACOUSTIC ||
                         p.op == OP_HOTSPOT2D || p.op == OP_GRADIENT || p.op == OP_SRAD) && same_extents(p);
  if (iterable && (p.op != OP_ACOUSTIC || n_state == 2)) {
    // WEIGHTED/HOTSPOT3D: state {X, scratch}; ACOUSTIC: state {prev, cur} plus
    // the two other workspace grids (two steps per pass where K2RA applies)
    float* state[4] = {pl->ws[0], pl->ws[1], pl->ws[2], pl->ws[3]};
    const float* aux[1] = {pl->ws[2]};
    int32_t ri = 0;
    const int ns = p.op == OP_ACOUSTIC ? 4 : 2;
    stencil_status s = stencil_iterate(pl, state, ns, aux, n_aux, n_steps, stream, &ri);
    if (s != STENCIL_OK) return s;
    result = state[ri];
  } else {
    if (n_steps != 1) return fail(STENCIL_E_UNSUPPORTED, "run_host: op is not iterable; use n_steps = 1");
    const float* in[2] = {pl->ws[0], n_state > 1 ? pl->ws[1] : (n_aux ? pl->ws[2] : nullptr)};
    int nin = op_arity(p.op);
    stencil_status s = stencil_apply(pl, in, nin, pl->ws[3], stream);
    if (s != STENCIL_OK) return s;
    result = pl->ws[3];
  }
  e = cudaMemcpyAsync(host_out, result, out_elems * sizeof(float), cudaMemcpyDeviceToHost, st);
  if (e != cudaSuccess) return cuda_fail(e, "D2H copy");
  e = cudaStreamSynchronize(st);
  if (e != cudaSuccess) return cuda_fail(e, "stream synchronize");
  return STENCIL_OK;
}

stencil_status stencil_run_host_batch(stencil_plan pl, const float* const* host_state, int32_t n_state,
                                      const float* const* host_aux, int32_t n_aux, int32_t n_steps,
                                      int32_t n_jobs, float* const* host_out) {
  if (!pl) return fail(STENCIL_E_INVALID, "NULL plan");
  if (!host_state || !host_out || n_state < 1 || n_state > 2 || n_aux < 0 || n_aux > 1 || n_jobs < 1 ||
      (n_aux > 0 && !host_aux))
    return fail(STENCIL_E_INVALID, "bad host buffers or counts");
  for (int32_t j = 0; j < n_jobs; ++j) {
    if (!host_out[j]) return fail(STENCIL_E_INVALID, "NULL host_out");
    for (int32_t s = 0; s < n_state; ++s)
      if (!host_state[j * n_state + s]) return fail(STENCIL_E_INVALID, "NULL host_state");
    for (int32_t a = 0; a < n_aux; ++a)
      if (!host_aux[j * n_aux + a]) return fail(STENCIL_E_INVALID, "NULL host_aux");
  }
  const StencilParams& p = pl->p;
  const bool iterable = (p.op == OP_WEIGHTED || p.op == OP_HOTSPOT3D || p.op == OP_ACOUSTIC ||
                         p.op == OP_HOTSPOT2D || p.op == OP_GRADIENT || p.op == OP_SRAD) && same_extents(p);
  if (!(iterable && (p.op != OP_ACOUSTIC || n_state == 2)) && n_steps != 1)
    return fail(STENCIL_E_UNSUPPORTED, "run_host_batch: op is not iterable; use n_steps = 1");
  DeviceGuard g(pl->device);
  if (g.err != cudaSuccess) return cuda_fail(g.err, "cudaSetDevice");
  const size_t in_elems = (size_t)(p.n[0] + 2 * p.ghost) * p.plane;
  const size_t out_elems = (size_t)(p.o[0] + 2 * p.ghost) * p.o[1] * p.o[2];
  const size_t elems = in_elems > out_elems ? in_elems : out_elems;
  constexpr int kSlots = 3, kGrids = 4;     // per slot: state0, state1, aux0 / spare, out / spare
  if (pl->wsb_elems < elems) {
    for (float* b : pl->wsb) cudaFree(b);
    pl->wsb.clear();
    pl->wsb_elems = 0;
    for (int i = 0; i < kSlots * kGrids; ++i) {
      float* b = nullptr;
      cudaError_t e = cudaMalloc(&b, elems * sizeof(float));
      if (e != cudaSuccess) return cuda_fail(e, "cudaMalloc (run_host_batch workspace)");
      pl->wsb.push_back(b);
    }
    pl->wsb_elems = elems;
  }
  // streams and events of this call
  cudaStream_t st_in = nullptr, st_comp = nullptr, st_out = nullptr;
  std::vector<cudaEvent_t> ev_in(n_jobs, nullptr), ev_comp(n_jobs, nullptr), ev_out(n_jobs, nullptr);
  struct Cleanup {
    cudaStream_t* s[3];
    std::vector<cudaEvent_t>* e[3];
    ~Cleanup() {
      // (an early error return must not leave copies into / out of the
      // caller's host buffers in flight)
      for (auto* x : s)
        if (*x) cudaStreamSynchronize(*x);
      for (auto* x : s)
        if (*x) cudaStreamDestroy(*x);
      for (auto* v : e)
        for (cudaEvent_t ev : *v)
          if (ev) cudaEventDestroy(ev);
    }
  } cleanup{{&st_in, &st_comp, &st_out}, {&ev_in, &ev_comp, &ev_out}};
  cudaError_t e = cudaStreamCreateWithFlags(&st_in, cudaStreamNonBlocking);
  if (e == cudaSuccess) e = cudaStreamCreateWithFlags(&st_comp, cudaStreamNonBlocking);
  if (e == cudaSuccess) e = cudaStreamCreateWithFlags(&st_out, cudaStreamNonBlocking);
  for (int32_t j = 0; j < n_jobs && e == cudaSuccess; ++j) {
    e = cudaEventCreateWithFlags(&ev_in[j], cudaEventDisableTiming);
    if (e == cudaSuccess) e = cudaEventCreateWithFlags(&ev_comp[j], cudaEventDisableTiming);
    if (e == cudaSuccess) e = cudaEventCreateWithFlags(&ev_out[j], cudaEventDisableTiming);
  }
  if (e != cudaSuccess) return cuda_fail(e, "run_host_batch: streams / events");
  for (int32_t j = 0; j < n_jobs; ++j) {
    float* const* slot = pl->wsb.data() + (j % kSlots) * kGrids;
    // copy in (after the slot's previous job has been copied out)
    if (j >= kSlots) {
      e = cudaStreamWaitEvent(st_in, ev_out[j - kSlots], 0);
      if (e != cudaSuccess) return cuda_fail(e, "run_host_batch: wait");
    }
    for (int32_t s = 0; s < n_state; ++s) {
      e = cudaMemcpyAsync(slot[s], host_state[j * n_state + s], in_elems * sizeof(float), cudaMemcpyHostToDevice,
                          st_in);
      if (e != cudaSuccess) return cuda_fail(e, "H2D copy");
    }
    for (int32_t a = 0; a < n_aux; ++a) {
      e = cudaMemcpyAsync(slot[2], host_aux[j * n_aux + a], in_elems * sizeof(float), cudaMemcpyHostToDevice, st_in);
      if (e != cudaSuccess) return cuda_fail(e, "H2D copy");
    }
    e = cudaEventRecord(ev_in[j], st_in);
    if (e == cudaSuccess) e = cudaStreamWaitEvent(st_comp, ev_in[j], 0);
    if (e != cudaSuccess) return cuda_fail(e, "run_host_batch: events");
    // compute
    const float* result = nullptr;
    if (iterable && (p.op != OP_ACOUSTIC || n_state == 2)) {
      float* state[4] = {slot[0], slot[1], slot[2], slot[3]};
      const float* aux[1] = {slot[2]};
      int32_t ri = 0;
      const int ns = p.op == OP_ACOUSTIC ? 4 : 2;
      stencil_status s = stencil_iterate(pl, state, ns, aux, n_aux, n_steps, st_comp, &ri);
      if (s != STENCIL_OK) return s;
      result = state[ri];
    } else {
      const float* in[2] = {slot[0], n_state > 1 ? slot[1] : (n_aux ? slot[2] : nullptr)};
      stencil_status s = stencil_apply(pl, in, op_arity(p.op), slot[3], st_comp);
      if (s != STENCIL_OK) return s;
      result = slot[3];
    }
    e = cudaEventRecord(ev_comp[j], st_comp);
    if (e == cudaSuccess) e = cudaStreamWaitEvent(st_out, ev_comp[j], 0);
    if (e != cudaSuccess) return cuda_fail(e, "run_host_batch: events");
    // copy out
    e = cudaMemcpyAsync(host_out[j], result, out_elems * sizeof(float), cudaMemcpyDeviceToHost, st_out);
    if (e != cudaSuccess) return cuda_fail(e, "D2H copy");
    e = cudaEventRecord(ev_out[j], st_out);
    if (e != cudaSuccess) return cuda_fail(e, "run_host_batch: events");
    // the next job's compute must not overwrite this slot before its copy-out:
    // slots are reused only kSlots jobs later, after ev_out (copy-in waits)
  }
  e = cudaStreamSynchronize(st_out);
  if (e == cudaSuccess) e = cudaStreamSynchronize(st_comp);
  if (e == cudaSuccess) e = cudaStreamSynchronize(st_in);
  if (e != cudaSuccess) return cuda_fail(e, "stream synchronize");
  return STENCIL_OK;
}

void stencil_plan_destroy(stencil_plan pl) {
  if (!pl) return;
  if (!pl->wsb.empty()) {
    DeviceGuard g(pl->device);
    for (float* b : pl->wsb) cudaFree(b);
  }
  if (!pl->ws.empty() || pl->srad_ws) {
    DeviceGuard g(pl->device);
    for (float* b : pl->ws) cudaFree(b);
    if (pl->srad_ws) cudaFree(pl->srad_ws);
  }
  delete pl;
}

}  // extern "C"
