// kernel_gather.cu — K5: WEIGHTED stencils of any shape through shared-memory
// tiles: strided slides (step > 1), even or asymmetric
// windows, 1D grids, wide boxes — every plan the TMA families (K1/K2/K3) do
// not take and K0 would otherwise run tap by tap from global memory.
//
// slide(size, step) of an output tile of OT = (OTZ, OTY, OTX)
// points reads the input box ((OT_d - 1) * step_d + size_d) per dimension —
// for a 2D 3x3 step-2 slide of a 16 x 128 tile, 33 x 257 floats, each read
// from HBM once instead of (size/step)^2 times.  The warps fill the box with
// coalesced 4-byte cp.async row copies, double-buffered so the next tile's box
// streams in while this one is evaluated (pad, is applied while
// loading: remapped index or the constant, so no padded copy exists); every thread
// evaluates its outputs from shared memory with the plan's non-zero taps in
// row-major order (or the separable row/column form) — exactly K0's sequence,
// so the two agree bitwise.  Slab mode (global z offset, ghost planes) and
// output regions along dimension 0 behave as in K0.
#include <cuda_runtime.h>

#include <algorithm>
#include <climits>
#include <cstdlib>
#include <mutex>
#include <string>

#include "common.cuh"
#include "launch.hpp"
#include "ops.cuh"
#include "tma.cuh"

namespace lift {
namespace {

constexpr int kThreads = 256;
constexpr int NJ = 4;                          // outputs per thread per pass
constexpr int NP = 2;                          // passes: tiles hold at most NP * NJ * kThreads outputs
constexpr int kMaxSmemFloats = 48 * 1024;     // 192 KiB box limit
constexpr int kMaxRows = 1024;                 // box rows (bz * by)

struct Tile {
  int otz, oty, otx;      // outputs per tile
  int bz, by, bx;         // input box; bx is the row pitch: the x extent wx + 3, rounded up to 4
  int wx;                 // x extent of the box the outputs read
};

__host__ __device__ inline Tile tile_of(const StencilParams& p, int otz, int oty, int otx) {
  Tile t{otz, oty, otx, 0, 0, 0, 0};
  t.bz = (otz - 1) * p.step[0] + p.size[0];
  t.by = (oty - 1) * p.step[1] + p.size[1];
  // box rows start at the tile's x origin rounded down to a multiple of 4
  // (up to 3 leading columns), so interior rows are copied in 16-byte pieces
  t.wx = (otx - 1) * p.step[2] + p.size[2];
  t.bx = (t.wx + 3 + 3) & ~3;
  return t;
}

// unpadded index -> in-grid index, or -1 for the constant (y / x dimensions)
__device__ __forceinline__ int64_t remap_or_const(int64_t i, int64_t n, int kind) {
  if (i >= 0 && i < n) return i;
  if (kind == PAD_CONSTANT) return -1;
  return pad_remap(i, n, kind);
}

// fill one box with 4-byte cp.async copies.  Warp w copies box rows w, w + 8,
// ...; pad per row is resolved first, one row per lane (element
// offset of the row's x origin in the input, or -1 for a value row, and the
// DAMPEN cells the row's y / z indices crossed), and handed to the copying
// lanes by shuffles — no shared table, no CTA barrier; x is remapped per
// element only on tiles touching the x edges.  Dimensions resolve innermost
// first, as in K0's fetch (x, then y, then z; reading A29 for DAMPEN), so the
// two kernels give the same bits.
__device__ __forceinline__ void fill_box(const StencilParams& p, const Tile& T, const float* __restrict__ in,
                                         float* dst_box, int64_t gz0, int64_t gy0, int64_t gx0, int warp,
                                         int lane) {
  constexpr int NWARP = kThreads / 32;
  const int nrows = T.bz * T.by;
  // row element b holds x = gxa + b: the origin gx0 rounded down to a multiple of 4
  const int sh = (int)(gx0 & 3);
  const int64_t gxa = gx0 - sh;
  const bool x_inside = gx0 >= 0 && gx0 + T.wx <= p.n[2];
  const int ncopy = sh + T.wx;      // columns the outputs read
  const bool quads = (p.n[2] % 4 == 0) && (reinterpret_cast<uintptr_t>(in) & 15u) == 0;
  const bool damp = has_dampen(p);
  for (int base = warp; base < nrows; base += NWARP * 32) {
    const int r = base + lane * NWARP;
    int64_t off = -1;
    int nrow = 0;
    if (r < nrows) {
      const int bzi = r / T.by, byi = r - bzi * T.by;
      int64_t iy = gy0 + byi;
      bool vrow = false;
      if (iy < 0 || iy >= p.n[1]) {
        if (p.kind[1] == PAD_CONSTANT) vrow = true;
        else {
          if (p.kind[1] == PAD_DAMPEN) nrow += (int)outside_dist(iy, p.n[1]);
          iy = pad_remap(iy, p.n[1], p.kind[1]);
        }
      }
      if (!vrow) {
        const int64_t gz = gz0 + bzi;
        const int64_t lz = plane_of(p, gz);
        if (lz >= 0) {
          if (p.kind[0] == PAD_DAMPEN) nrow += (int)outside_dist(gz, p.gnz);
          off = lz * p.plane + iy * p.row + (x_inside ? gxa : 0);
        }
      } else {
        nrow = 0;       // the y value cell: only x's DAMPEN cells (inside it) count
      }
    }
    const int cnt = min(32, (nrows - base + NWARP - 1) / NWARP);
    for (int i = 0; i < cnt; ++i) {
      const int64_t o = __shfl_sync(0xffffffffu, off, i);
      const int nr = __shfl_sync(0xffffffffu, nrow, i);
      float* dst = dst_box + (base + i * NWARP) * T.bx;
      if (!damp) {
        if (o < 0) {
          for (int b = lane; b < T.bx; b += 32) dst[b] = p.pad_value;
        } else if (x_inside) {
          const float* s0 = in + o;
          if (quads && (reinterpret_cast<uintptr_t>(s0) & 15u) == 0) {
            // gxa and nx are multiples of 4 and gx0 + wx <= nx: the last quad ends in the row
            for (int b = 4 * lane; b < ncopy; b += 128) cp_async16(dst + b, s0 + b);
          } else {
            for (int b = lane; b < ncopy; b += 32) cp_async4(dst + b, s0 + b);
          }
        } else {
          // a tile touching the x edges: the in-grid columns [blo, bhi) of the
          // row are copied like an interior row (16-byte pieces: gxa and nx are
          // multiples of 4, so the range is quad-aligned), only the
          // out-of-grid columns are remapped one by one
          const int64_t nx = p.n[2];
          const int blo = (int)(gxa < 0 ? -gxa : 0);
          const int64_t hi_ = nx - gxa < (int64_t)T.bx ? nx - gxa : (int64_t)T.bx;
          const int bhi = hi_ > blo ? (int)hi_ : blo;
          const float* s0 = in + o + gxa;
          if (quads) {
            for (int b = blo + 4 * lane; b < bhi; b += 128) cp_async16(dst + b, s0 + b);
          } else {
            for (int b = blo + lane; b < bhi; b += 32) cp_async4(dst + b, s0 + b);
          }
          for (int b = lane; b < blo + (T.bx - bhi); b += 32) {
            const int bb = b < blo ? b : bhi + (b - blo);
            const int64_t ix = remap_or_const(gxa + bb, nx, p.kind[2]);
            if (ix < 0) dst[bb] = p.pad_value;
            else cp_async4(dst + bb, in + o + ix);
          }
        }
      } else {
        // DAMPEN plans: values computed directly (decay^k scaling)
        for (int b = lane; b < T.bx; b += 32) {
          int64_t ix = gxa + b;
          int k = nr;
          float v;
          if ((ix < 0 || ix >= p.n[2]) && p.kind[2] == PAD_CONSTANT) {
            v = p.pad_value;
            k = 0;
          } else {
            if (ix < 0 || ix >= p.n[2]) {
              if (p.kind[2] == PAD_DAMPEN) k += (int)outside_dist(ix, p.n[2]);
              ix = pad_remap(ix, p.n[2], p.kind[2]);
            }
            v = o < 0 ? p.pad_value : __ldg(in + o + (x_inside ? ix - gxa : ix));
          }
          dst[b] = k ? __fmul_rn(v, dampen_pow(p.pad_decay, k)) : v;
        }
      }
    }
  }
}

// nbuf = 2: the next tile's box streams in (cp.async) while this one is evaluated.
// SZ, SY, SX > 0: compile-time window (all taps non-zero, or separable 2D)
template <int SZ, int SY, int SX>
__global__ void __launch_bounds__(kThreads, 3) k5_gather(const __grid_constant__ StencilParams p, Tile T,
                                                      const float* __restrict__ in, float* __restrict__ out,
                                                      int64_t ntz, int64_t nty, int64_t ntx, int nbuf,
                                                      const __grid_constant__ CUtensorMap tmap, int use_tma) {
  extern __shared__ __align__(128) float box[];
  __shared__ int toff[kMaxTaps];
  __shared__ uint64_t tbar[2];
  pdl_launch_dependents();
  const int BYX = T.by * T.bx;
  const int box_floats = T.bz * BYX;
  const int buf_floats = (box_floats + 31) & ~31;     // buffers 128-B aligned (TMA destinations)
  for (int t = threadIdx.x; t < p.ntaps; t += kThreads)
    toff[t] = p.tap[t][0] * BYX + p.tap[t][1] * T.bx + p.tap[t][2];
  if (threadIdx.x == 0) {
    mbar_init(&tbar[0], 1);
    mbar_init(&tbar[1], 1);
    fence_mbar_init();
    if (use_tma) prefetch_tmap(&tmap);
  }
  __syncthreads();
  pdl_wait();
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int64_t oz_n = p.reg1 - p.reg0, oy_n = p.o[1], ox_n = p.o[2];
  const int64_t out_plane = p.o[1] * p.o[2];
  const int64_t ntiles = ntz * nty * ntx;
  const int nout = T.otz * T.oty * T.otx;
  auto origin = [&](int64_t tile, int64_t& oz0, int64_t& oy0, int64_t& ox0) {
    // 32-bit division: ntiles < 2^31 (checked at launch)
    const uint32_t t32 = (uint32_t)tile, r = t32 / (uint32_t)ntx;
    const uint32_t tx = t32 - r * (uint32_t)ntx;
    const uint32_t tz = r / (uint32_t)nty, ty = r - tz * (uint32_t)nty;
    // widen before multiplying: a 1D plan's x extent may exceed 2^32
    oz0 = p.reg0 + (int64_t)tz * T.otz;
    oy0 = (int64_t)ty * T.oty;
    ox0 = (int64_t)tx * T.otx;
  };
  // Interior boxes (every cell the outputs read inside the grid, so no pad)
  // arrive as ONE TMA box load issued by one thread (use_tma: 16-B aligned
  // rows, box dims <= 256); edge boxes are filled by the warps (fill_box).
  // tma_mask / tma_phase: per buffer, whether its pending fill is a TMA load
  // and the parity of its barrier.
  unsigned tma_mask = 0u, tma_phase = 0u;      // bit b: buffer b (no local-memory arrays)
  auto fill = [&](int64_t tile, int buf) {
    int64_t oz0, oy0, ox0;
    origin(tile, oz0, oy0, ox0);
    // unpadded coordinates of the box origin (global z)
    const int64_t gz0 = p.z_off + oz0 * p.step[0] - p.lo[0], gy0 = oy0 * p.step[1] - p.lo[1];
    const int64_t gx0 = ox0 * p.step[2] - p.lo[2];
    const int64_t lz0 = gz0 - p.z_off + p.ghost;
    const bool interior = use_tma && gx0 >= 0 && gx0 + T.wx <= p.n[2] && gy0 >= 0 && gy0 + T.by <= p.n[1] &&
                          gz0 >= 0 && gz0 + T.bz <= p.gnz && lz0 >= 0 && lz0 + T.bz <= p.n[0] + 2 * p.ghost;
    tma_mask = interior ? (tma_mask | (1u << buf)) : (tma_mask & ~(1u << buf));
    if (interior) {
      if (threadIdx.x == 0) {
        fence_proxy_async_smem();     // the buffer's earlier generic-proxy accesses before the async-proxy write
        mbar_arrive_expect_tx(&tbar[buf], (uint32_t)(box_floats * 4));
        tma_load_3d(box + buf * buf_floats, &tmap, &tbar[buf], (int)(gx0 & ~(int64_t)3), (int)gy0, (int)lz0);
      }
    } else {
      fill_box(p, T, in, box + buf * buf_floats, gz0, gy0, gx0, warp, lane);
    }
    cp_async_commit();                // (an empty group for a TMA fill keeps the group count per tile)
  };
  auto wait_tma = [&](int buf) {
    if ((tma_mask >> buf) & 1u) {
      mbar_wait(&tbar[buf], (tma_phase >> buf) & 1u);
      tma_phase ^= 1u << buf;
    }
  };
  // this thread's outputs within a tile (tile-invariant: no per-tile division):
  // k = tid + (pass * NJ + j) * kThreads, at most NP passes (nout <= NP*NJ*kThreads)
  int woff[NP * NJ], kxs[NP * NJ], kys[NP * NJ], kzs[NP * NJ];
#pragma unroll
  for (int q = 0; q < NP * NJ; ++q) {
    const int k = threadIdx.x + q * kThreads;
    const int kx = k % T.otx, kr = k / T.otx;
    const int ky = kr % T.oty, kz = kr / T.oty;
    const bool v = k < nout;
    kxs[q] = kx;
    kys[q] = ky;
    kzs[q] = v ? kz : INT32_MAX / 2;     // invalid slots fail the range check below
    woff[q] = v ? kz * p.step[0] * BYX + ky * p.step[1] * T.bx + kx * p.step[2] : 0;
  }
  int cur = 0;
  if ((int64_t)blockIdx.x < ntiles) fill(blockIdx.x, 0);
  for (int64_t tile = blockIdx.x; tile < ntiles; tile += gridDim.x) {
    const int64_t next = tile + gridDim.x;
    float* bcur = box + cur * buf_floats;
    if (nbuf == 2) {
      if (next < ntiles) fill(next, cur ^ 1);
      else cp_async_commit();
      cp_async_wait<1>();
    } else {
      cp_async_wait<0>();
    }
    wait_tma(cur);
    __syncthreads();
    int64_t oz0, oy0, ox0;
    origin(tile, oz0, oy0, ox0);
    const int xsh = (int)((ox0 * p.step[2] - p.lo[2]) & 3);   // leading columns of the aligned box rows
    // each thread evaluates NJ outputs per pass: the tap loop's index / weight
    // loads are shared by NJ independent FMA chains
#pragma unroll
    for (int ps = 0; ps < NP; ++ps) {
      if (threadIdx.x + ps * NJ * kThreads >= nout) continue;   // (no break: keeps the loop fully unrolled)
      int64_t oidx[NJ];
      bool ok[NJ];
#pragma unroll
      for (int j = 0; j < NJ; ++j) {
        const int q = ps * NJ + j;
        const int64_t oz = oz0 + kzs[q], oy = oy0 + kys[q], ox = ox0 + kxs[q];
        ok[j] = oz - p.reg0 < oz_n && oy < oy_n && ox < ox_n;
        oidx[j] = (oz + p.ghost) * out_plane + oy * ox_n + ox;
      }
      float acc[NJ];
#pragma unroll
      for (int j = 0; j < NJ; ++j) acc[j] = 0.0f;
      const float* wj[NJ];
#pragma unroll
      for (int j = 0; j < NJ; ++j) wj[j] = bcur + xsh + woff[ps * NJ + j];
      if constexpr (SZ > 0) {
        // compile-time window (dense weights or separable 2D): unrolled taps,
        // immediate x offsets, the same operation order as the tap list
        if (p.sep) {
#pragma unroll
          for (int a = 0; a < SY; ++a) {
            float h[NJ];
#pragma unroll
            for (int j = 0; j < NJ; ++j) h[j] = 0.0f;
#pragma unroll
            for (int b = 0; b < SX; ++b) {
              const float wv = p.sv[b];
#pragma unroll
              for (int j = 0; j < NJ; ++j) h[j] = __fmaf_rn(wv, wj[j][a * T.bx + b], h[j]);
            }
            const float wu = p.su[a];
#pragma unroll
            for (int j = 0; j < NJ; ++j) acc[j] = __fmaf_rn(wu, h[j], acc[j]);
          }
        } else {
          // even x step: every output's window starts at the same parity (xsh's), so
          // tap pairs starting on an even column load as one 8-byte LDS; the FMA
          // order is the tap list's either way
          auto dense = [&](auto PARC) {
            constexpr int PAR = decltype(PARC)::value;
#pragma unroll
            for (int kz = 0; kz < SZ; ++kz)
#pragma unroll
              for (int ky = 0; ky < SY; ++ky) {
                const int ro = kz * BYX + ky * T.bx;
                static_for<SX>([&](auto KX) {
                  constexpr int kx = decltype(KX)::value;
                  const float* wr = p.w + (kz * SY + ky) * SX;
                  if constexpr (PAR >= 0 && (kx + PAR) % 2 == 0 && kx + 1 < SX) {
#pragma unroll
                    for (int j = 0; j < NJ; ++j) {
                      const float2 v = *reinterpret_cast<const float2*>(wj[j] + ro + kx);
                      acc[j] = __fmaf_rn(wr[kx], v.x, acc[j]);
                      acc[j] = __fmaf_rn(wr[kx + 1], v.y, acc[j]);
                    }
                  } else if constexpr (PAR >= 0 && (kx + PAR) % 2 == 1 && kx > 0) {
                    // second tap of a pair: done above
                  } else {
#pragma unroll
                    for (int j = 0; j < NJ; ++j) acc[j] = __fmaf_rn(wr[kx], wj[j][ro + kx], acc[j]);
                  }
                });
              }
          };
          if (p.step[2] % 2 == 0) {
            if (xsh & 1) dense(std::integral_constant<int, 1>{});
            else dense(std::integral_constant<int, 0>{});
          } else {
            dense(std::integral_constant<int, -1>{});
          }
        }
      } else if (p.sep) {
        // separable 2D weights: rows first (x taps in order), then the column (K0's order)
        for (int a = 0; a < p.size[1]; ++a) {
          float h[NJ];
#pragma unroll
          for (int j = 0; j < NJ; ++j) h[j] = 0.0f;
          for (int b = 0; b < p.size[2]; ++b) {
            const float wv = p.sv[b];
            const int o = a * T.bx + b;
#pragma unroll
            for (int j = 0; j < NJ; ++j) h[j] = __fmaf_rn(wv, wj[j][o], h[j]);
          }
          const float wu = p.su[a];
#pragma unroll
          for (int j = 0; j < NJ; ++j) acc[j] = __fmaf_rn(wu, h[j], acc[j]);
        }
      } else {
        for (int t = 0; t < p.ntaps; ++t) {
          const float wv = p.w[t];
          const int o = toff[t];
#pragma unroll
          for (int j = 0; j < NJ; ++j) acc[j] = __fmaf_rn(wv, wj[j][o], acc[j]);
        }
      }
#pragma unroll
      for (int j = 0; j < NJ; ++j)
        if (ok[j]) out[oidx[j]] = acc[j];
    }
    __syncthreads();     // bcur is refilled two tiles from now
    if (nbuf == 2) {
      cur ^= 1;
    } else if (next < ntiles) {
      fill(next, 0);
    }
  }
}

struct Shape {
  int otz, oty, otx;
};

// output tile per dimensionality: 3D (2, 4, 128), 2D (1, 16, 128), 1D (1, 1, 1024),
// halved (largest first) until the box fits
bool choose(const StencilParams& p, Tile* T, bool tma = false) {
  const bool d3 = p.o[0] > 1 || p.size[0] > 1;
  const bool d2 = p.o[1] > 1 || p.size[1] > 1;
  // 3D: long box rows amortise the per-row work of the fill (measured on 512^3
  // step-2 slides: (2, 4, 128) 1217 GB/s vs (4, 8, 32) 903 GB/s for 3x3x3)
  Shape s = d3 ? Shape{2, 4, 128} : (d2 ? Shape{1, 16, 128} : Shape{1, 1, 1024});
  if (d3) {
    if (const char* e = getenv("LIFT_K5_3D")) {     // A/B hook: 1 = (2, 8, 64), 2 = (1, 8, 128), 3 = (4, 8, 32)
      const int v = atoi(e);
      if (v == 1) s = Shape{2, 8, 64};
      if (v == 2) s = Shape{1, 8, 128};
      if (v == 3) s = Shape{4, 8, 32};
    }
  }
  // TMA boxes are at most 256 per dimension: narrower, taller tiles (3D
  // (2, 8, 64), 2D (1, 32, 64)) — with the fill in one instruction there is no
  // per-row cost to amortise
  if (tma) {
    if (d3) s = Shape{2, 8, 64};
    else if (d2) s = Shape{1, 32, 64};
    if (const char* e = getenv("LIFT_K5_TMA_SHAPE")) {   // A/B hook
      const int v = atoi(e);
      if (v == 1) s = d3 ? Shape{2, 4, 124} : Shape{1, 16, 124};
      if (v == 2) s = d3 ? Shape{4, 8, 32} : Shape{1, 64, 32};
      if (v == 3) s = d3 ? Shape{1, 16, 64} : Shape{1, 16, 64};
      if (v == 4) s = d3 ? Shape{2, 16, 32} : Shape{1, 32, 32};
    }
  }
  for (int it = 0; it < 24; ++it) {
    const Tile t = tile_of(p, s.otz, s.oty, s.otx);
    const bool tma_fits = !tma || (t.bx <= 256 && t.by <= 256 && t.bz <= 256);
    if ((int64_t)t.bz * t.by * t.bx <= kMaxSmemFloats && s.otz * s.oty * s.otx <= NP * NJ * kThreads &&
        t.bz * t.by <= kMaxRows && tma_fits) {
      *T = t;
      return true;
    }
    if (s.otx >= 2 * s.oty && s.otx > 1) s.otx /= 2;
    else if (s.oty > 1) s.oty /= 2;
    else if (s.otz > 1) s.otz /= 2;
    else if (s.otx > 1) s.otx /= 2;
    else return false;
  }
  return false;
}

}  // namespace

bool gather_supported(const StencilParams& p) {
  if (p.op != OP_WEIGHTED || p.ntaps < 1) return false;
  Tile t;
  return choose(p, &t);
}

cudaError_t launch_gather(const StencilParams& p, const float* in0, float* out, cudaStream_t stream, int num_sms,
                          std::string* err) {
  // TMA box fills for the interior tiles: 16-B aligned rows (nx % 4 == 0, an
  // aligned base); LIFT_K5_TMA=0 keeps the cp.async fill everywhere (A/B)
  // (measured, profiles/r02_k5_tma.txt: 2D windows and 3D windows of depth <= 2
  // gain 36-62%; the 3x3x3 box is compute-bound and runs faster on the
  // cp.async path's (2, 4, 128) tiles than on any TMA-sized tile)
  const char* et = getenv("LIFT_K5_TMA");
  const bool deep3d = (p.o[0] > 1 || p.size[0] > 1) && p.size[0] >= 3;
  bool tma = !(et && et[0] == '0') && (!deep3d || (et && et[0] == '1')) && p.n[2] % 4 == 0 &&
             (reinterpret_cast<uintptr_t>(in0) & 15u) == 0;
  Tile T;
  if (!(tma && choose(p, &T, true))) {
    tma = false;
    if (!choose(p, &T)) {
      *err = "gather: window box exceeds shared memory";
      return cudaErrorInvalidConfiguration;
    }
  }
  CUtensorMap tmap{};
  if (tma && !encode_tensor_map_3d(&tmap, in0, p.n[2], p.n[1], p.n[0] + 2 * p.ghost, (uint32_t)T.bx, (uint32_t)T.by,
                                   (uint32_t)T.bz, err))
    return cudaErrorInvalidValue;
  const int64_t oz_n = p.reg1 - p.reg0;
  if (oz_n <= 0 || p.o[1] <= 0 || p.o[2] <= 0) return cudaSuccess;
  const int64_t ntz = (oz_n + T.otz - 1) / T.otz, nty = (p.o[1] + T.oty - 1) / T.oty;
  const int64_t ntx = (p.o[2] + T.otx - 1) / T.otx;
  const size_t box_bytes = (size_t)(((int64_t)T.bz * T.by * T.bx + 31) & ~31ll) * sizeof(float);
  const int nbuf = 2 * box_bytes <= (size_t)kMaxSmemFloats * 4 ? 2 : 1;
  const size_t smem = nbuf * box_bytes;
  // compile-time windows for the common shapes when every tap is non-zero
  // (the unrolled loop then runs the tap list's order) or the weights are separable
  const int sz = p.size[0], sy = p.size[1], sx = p.size[2];
  const bool dense = p.ntaps == sz * sy * sx;
  const bool ok = (dense || p.sep) && !getenv("LIFT_K5_GENERIC");
  const void* fn = reinterpret_cast<const void*>(&k5_gather<0, 0, 0>);
  if (ok && sz == 1 && sy == 3 && sx == 3) fn = reinterpret_cast<const void*>(&k5_gather<1, 3, 3>);
  else if (ok && sz == 1 && sy == 5 && sx == 5) fn = reinterpret_cast<const void*>(&k5_gather<1, 5, 5>);
  else if (ok && sz == 1 && sy == 2 && sx == 2) fn = reinterpret_cast<const void*>(&k5_gather<1, 2, 2>);
  else if (dense && !getenv("LIFT_K5_GENERIC") && sz == 3 && sy == 3 && sx == 3)
    fn = reinterpret_cast<const void*>(&k5_gather<3, 3, 3>);
  else if (dense && !getenv("LIFT_K5_GENERIC") && sz == 2 && sy == 2 && sx == 2)
    fn = reinterpret_cast<const void*>(&k5_gather<2, 2, 2>);
  static std::once_flag once;
  std::call_once(once, [] {
    for (const void* f : {reinterpret_cast<const void*>(&k5_gather<0, 0, 0>), reinterpret_cast<const void*>(&k5_gather<1, 3, 3>),
                          reinterpret_cast<const void*>(&k5_gather<1, 5, 5>), reinterpret_cast<const void*>(&k5_gather<1, 2, 2>),
                          reinterpret_cast<const void*>(&k5_gather<3, 3, 3>), reinterpret_cast<const void*>(&k5_gather<2, 2, 2>)})
      cudaFuncSetAttribute(f, cudaFuncAttributeMaxDynamicSharedMemorySize, kMaxSmemFloats * 4);
  });
  int occ = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, fn, kThreads, smem) != cudaSuccess || occ < 1) occ = 1;
  cudaGetLastError();
  int64_t grid = (int64_t)num_sms * occ;
  const int64_t ntiles = ntz * nty * ntx;
  if (ntiles >= (1ll << 31)) {
    *err = "gather: too many tiles";
    return cudaErrorInvalidConfiguration;
  }
  if (grid > ntiles) grid = ntiles;
  const bool fz = p.put_lo || p.put_hi || p.fused_step || p.wait_lo || p.wait_hi;
  int nb = nbuf, ut = tma ? 1 : 0;
  void* args[] = {(void*)&p,   (void*)&T,   (void*)&in0, (void*)&out, (void*)&ntz,
                  (void*)&nty, (void*)&ntx, (void*)&nb,  (void*)&tmap, (void*)&ut};
  set_last_kernel(tma ? "k5_gather (TMA)" : "k5_gather");
  return launch_kernel(fn, dim3((unsigned)grid), dim3(kThreads), args, smem, stream, !fz);
}

}  // namespace lift
