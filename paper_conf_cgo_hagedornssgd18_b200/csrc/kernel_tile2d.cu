// kernel_tile2d.cu — K1: the 2D stencil on TMA-staged halo'd tiles.
//
// map_2(f, slide_2(size, step, pad_2(...))) over a 2D
// grid.  The output is cut into 128 x 48 tiles (overlapped tiling, P:693-822:
// each tile's input box carries the 2R-wide overlap).  Persistent CTAs (one
// wave: grid = SMs x resident CTAs) take tiles with a grid stride, so in every
// round the CTAs cover a band of consecutive tiles in row-major order and the
// overlap rows/columns of neighbouring tiles come from L2.  Per CTA an elected
// producer thread streams each tile's box ((128+8) x (48+2RY) floats per input
// grid) into a 2-stage shared-memory ring with TMA and mbarriers; 8 consumer
// warps each sweep 6 output rows down the box.  Every box row is read from
// shared memory once per warp (one LDS.128 per lane; the in-row neighbours
// come from the adjacent lanes by warp shuffles) and immediately added to the
// 2RY+1 output rows in flight, so each output's FMA chain runs in row-major
// tap order — the order K0 uses.  Separable weights (the binomial Gaussian)
// take the row sum once per box row and then one FMA per output row
// (10 instead of 25 FMA per point), star weights skip the off-axis taps.
// 4 outputs per lane leave as one st.global.v4.  Edge tiles rewrite their
// out-of-grid halo cells (halo.cuh) before use.
#include <cuda.h>
#include <cuda_runtime.h>

#include <cstdlib>
#include <climits>
#include <mutex>
#include <string>

#include "common.cuh"
#include "halo.cuh"
#include "launch.hpp"
#include "ops.cuh"
#include "tma.cuh"

namespace lift {
namespace {

constexpr int TX = 128;
constexpr int XH = 4;
constexpr int BX = TX + 2 * XH;
constexpr int NW = 8;
constexpr int kSradMaxParts = 2048;     // q0 partials one K1S pass can reduce (8 per consumer thread)
constexpr int NCONS = NW * 32;
constexpr unsigned FULL = 0xffffffffu;

enum K1Op { K1_WBOX = 0, K1_SRAD1 = 1, K1_SRAD2 = 2, K1_WSTAR = 3, K1_WSEP = 4, K1_HOT2D = 5, K1_GRAD = 6 };

template <int RY, int RPW, int S, int NIN>
struct Cfg {
  static constexpr int TY = NW * RPW;
  static constexpr int BY = TY + 2 * RY;
  static constexpr int BOX_BYTES = BX * BY * 4;
  static constexpr int BOX_FLOATS = ((BOX_BYTES + 127) / 128) * 128 / 4;
  static constexpr int STAGE_FLOATS = NIN * BOX_FLOATS;
  static constexpr int SMEM = S * STAGE_FLOATS * 4 + 2 * S * 8 + 128;
};

// x-window of one box row for the 4 outputs of a lane: offsets -RX .. 3+RX
// (centre float4 from shared memory, neighbours from the adjacent lanes)
template <int RX>
__device__ __forceinline__ void load_row(const float4* row4, int lane, float (&xw)[4 + 2 * RX]) {
  const float4 c = row4[XH / 4 + lane];
  const float4 e = row4[lane == 0 ? 0 : (TX + XH) / 4];
  const float cv[4] = {c.x, c.y, c.z, c.w};
  const float ev[4] = {e.x, e.y, e.z, e.w};
#pragma unroll
  for (int k = 1; k <= RX; ++k) {
    float l = __shfl_up_sync(FULL, cv[4 - k], 1);     // x - k from the left lane
    float r = __shfl_down_sync(FULL, cv[k - 1], 1);   // x + 3 + k from the right lane
    if (lane == 0) l = ev[4 - k];
    if (lane == 31) r = ev[k - 1];
    xw[RX - k] = l;
    xw[RX + 3 + k] = r;
  }
#pragma unroll
  for (int i = 0; i < 4; ++i) xw[RX + i] = cv[i];
}

// Accessor over a ring of x-windows (SRAD): rows[DY + RY][I + RX + DX].
template <int RY, int RX, int I>
struct RingAcc {
  const float (*rows)[4 + 2 * RX];
  template <int DZ, int DY, int DX>
  __device__ __forceinline__ float at() const {
    static_assert(DZ == 0, "2D");
    return rows[DY + RY][I + RX + DX];
  }
};

template <int OP, int RY, int RX, int RPW, int S, int NIN, int MINB, bool LDG>
__global__ void __launch_bounds__(NCONS + 32, MINB)
    k1_tile(const __grid_constant__ StencilParams p, const __grid_constant__ CUtensorMap map0,
            const __grid_constant__ CUtensorMap map1, const float* __restrict__ src0,
            const float* __restrict__ src1, float* __restrict__ out, int ntx, int nty) {
  using C = Cfg<RY, RPW, S, NIN>;
  constexpr int TY = C::TY;
  constexpr int W = 4 + 2 * RX;
  constexpr int SY = 2 * RY + 1, SX = 2 * RX + 1;
  constexpr int BX4 = BX / 4;
  constexpr int SF4 = C::STAGE_FLOATS / 4;
  constexpr int BF4 = C::BOX_FLOATS / 4;
  extern __shared__ __align__(128) float4 dsm4[];
  uint64_t* full = reinterpret_cast<uint64_t*>(dsm4 + S * SF4);
  uint64_t* empty = full + S;

  // strided tile assignment: in round k all CTAs work on tiles
  // [k*grid, (k+1)*grid) of the row-major tile order, so the tiles above and
  // below (whose rows are this tile's halo) are in flight in the same or the
  // neighbouring round and the overlap comes from L2
  const int64_t ntiles = (int64_t)ntx * nty;
  const int nt = (int)((ntiles - blockIdx.x + gridDim.x - 1) / gridDim.x);
  if (nt <= 0) return;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;

  if (threadIdx.x == 0) {
    for (int s = 0; s < S; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NW);
    }
    fence_mbar_init();
  }
  __syncthreads();
  pdl_launch_dependents();   // PDL: let the next launch ramp up now
  pdl_wait();                // ... and wait for the previous one before any global access

  if (warp == NW) {
    if (!LDG && lane == 0) {
      prefetch_tmap(&map0);
      if (NIN > 1) prefetch_tmap(&map1);
      int s = 0;
      uint32_t pass = 0;
      for (int i = 0; i < nt; ++i) {
        if (pass > 0) mbar_wait(&empty[s], (pass - 1) & 1);
        const int64_t t = blockIdx.x + (int64_t)i * gridDim.x;
        const int x0 = (int)(t % ntx) * TX, y0 = (int)(t / ntx) * TY;
        mbar_arrive_expect_tx(&full[s], NIN * C::BOX_BYTES);
        tma_load_3d(dsm4 + s * SF4, &map0, &full[s], x0 - XH, y0 - RY, 0);
        if constexpr (NIN > 1) tma_load_3d(dsm4 + s * SF4 + BF4, &map1, &full[s], x0 - XH, y0 - RY, 0);
        if (++s == S) { s = 0; ++pass; }
      }
    }
    return;
  }

  const int nx = (int)p.n[2], ny = (int)p.n[1];
  const bool zero_fill_ok = p.pad_value == 0.0f && p.kind[1] == PAD_CONSTANT && p.kind[2] == PAD_CONSTANT;
  const int r0 = warp * RPW;   // first output row of this warp (tile-relative)
  // 128-bit stores need 16-B aligned rows (nx % 4 == 0 and an aligned base)
  const bool vec = (nx % 4 == 0) && ((reinterpret_cast<uintptr_t>(out) & 15u) == 0);
  auto fixup = [&](int s, int x0, int y0) {
    const bool edge = (x0 == 0) || (x0 + TX + RX > nx) || (y0 < RY) || (y0 + TY + RY > ny);
    if (edge && !zero_fill_ok) {
      fixup_tile<RY, RX, XH, BX, C::BY, NCONS>(p, reinterpret_cast<float*>(dsm4 + s * SF4), src0, 0, x0, y0,
                                               threadIdx.x);
      if constexpr (NIN > 1)
        fixup_tile<RY, RX, XH, BX, C::BY, NCONS>(p, reinterpret_cast<float*>(dsm4 + s * SF4 + BF4), src1, 0, x0,
                                                 y0, threadIdx.x);
      fence_proxy_async_smem();
      named_bar_sync(1, NCONS);
    }
  };
  auto compute = [&](int s, int x0, int y0) {
    const int xo = x0 + 4 * lane;
    const bool x_ok = xo < nx;
    const float4* box0 = dsm4 + s * SF4 + r0 * BX4;     // box row r0 = output row r0 - RY
    float* orow = out + ((int64_t)(y0 + r0) * nx + xo);
    auto store = [&](int o, const float (&v)[4]) {
      if (!(x_ok && y0 + r0 + o < ny)) return;
      float* dst = orow + (int64_t)o * nx;
      if (vec) {
        stg128(dst, make_float4(v[0], v[1], v[2], v[3]));
      } else {
#pragma unroll
        for (int q = 0; q < 4; ++q)
          if (xo + q < nx) dst[q] = v[q];
      }
    };

    if constexpr (OP == K1_WBOX || OP == K1_WSTAR || OP == K1_WSEP) {
      // Box rows stream in top to bottom; each row adds its taps to the 2RY+1
      // outputs in flight, so every output's chain runs in row-major tap order.
      float acc[SY][4];
      static_for<RPW + 2 * RY>([&](auto KR) {
        constexpr int kr = decltype(KR)::value;
        float xw[W];
        load_row<RX>(box0 + kr * BX4, lane, xw);
        float h[4];
        if constexpr (OP == K1_WSEP) {
#pragma unroll
          for (int q = 0; q < 4; ++q) {
            float a = 0.0f;
#pragma unroll
            for (int kx = 0; kx < SX; ++kx) a = __fmaf_rn(p.sv[kx], xw[q + kx], a);
            h[q] = a;
          }
        }
        static_for<SY>([&](auto KY) {
          constexpr int ky = decltype(KY)::value;
          constexpr int o = kr - ky;                  // output row (warp-relative) this box row feeds
          if constexpr (o >= 0 && o < RPW) {
            constexpr int slot = o % SY;
#pragma unroll
            for (int q = 0; q < 4; ++q) {
              float a = ky == 0 ? 0.0f : acc[slot][q];
              if constexpr (OP == K1_WSEP) {
                a = __fmaf_rn(p.su[ky], h[q], a);
              } else if constexpr (OP == K1_WSTAR) {
                if constexpr (ky == RY) {
#pragma unroll
                  for (int kx = 0; kx < SX; ++kx) a = __fmaf_rn(p.wbox[ky * SX + kx], xw[q + kx], a);
                } else {
                  a = __fmaf_rn(p.wbox[ky * SX + RX], xw[q + RX], a);
                }
              } else {
#pragma unroll
                for (int kx = 0; kx < SX; ++kx) a = __fmaf_rn(p.wbox[ky * SX + kx], xw[q + kx], a);
              }
              acc[slot][q] = a;
            }
            if constexpr (ky == 2 * RY) store(o, acc[slot]);
          }
        });
      });
    } else {
      // SRAD: all taps of an output at once from a ring of 2RY+1 x-windows
      float ra[SY][W];
      float rb[(NIN > 1) ? SY : 1][W];
      static_for<RPW + 2 * RY>([&](auto KR) {
        constexpr int kr = decltype(KR)::value;
        constexpr int slot = kr % SY;
        load_row<RX>(box0 + kr * BX4, lane, ra[slot]);
        if constexpr (NIN > 1) load_row<RX>(box0 + BF4 + kr * BX4, lane, rb[slot]);
        constexpr int o = kr - 2 * RY;
        if constexpr (o >= 0) {
          // rows o .. o+2RY of the box sit in slots (o + k) % SY
          float wa[SY][W], wb[(NIN > 1) ? SY : 1][W];
#pragma unroll
          for (int k = 0; k < SY; ++k)
#pragma unroll
            for (int q = 0; q < W; ++q) {
              wa[k][q] = ra[(o + k) % SY][q];
              if constexpr (NIN > 1) wb[k][q] = rb[(o + k) % SY][q];
            }
          float v[4];
          static_for<4>([&](auto I) {
            constexpr int ii = decltype(I)::value;
            if constexpr (OP == K1_SRAD1) {
              v[ii] = op_srad1(RingAcc<RY, RX, ii>{wa}, p.prm);
            } else if constexpr (OP == K1_GRAD) {
              v[ii] = op_gradient(RingAcc<RY, RX, ii>{wa}, p.prm);
            } else if constexpr (OP == K1_HOT2D) {
              v[ii] = op_hotspot2d(RingAcc<RY, RX, ii>{wa}, RingAcc<RY, RX, ii>{wb}, p.prm);   // (T, P)
            } else {
              v[ii] = op_srad2(RingAcc<RY, RX, ii>{wa}, RingAcc<RY, RX, ii>{wb}, p.prm);   // (c, I)
            }
          });
          store(o, v);
        }
      });
    }
  };

  if constexpr (!LDG) {
    int s = 0;
    uint32_t pass = 0;
    for (int i = 0; i < nt; ++i) {
      mbar_wait(&full[s], pass & 1);
      const int64_t t = blockIdx.x + (int64_t)i * gridDim.x;
      const int x0 = (int)(t % ntx) * TX, y0 = (int)(t / ntx) * TY;
      fixup(s, x0, y0);
      compute(s, x0, y0);
      __syncwarp();
      if (lane == 0) mbar_arrive(&empty[s]);
      if (++s == S) { s = 0; ++pass; }
    }
  } else {
    // rows that TMA cannot describe (nx % 4 != 0 or an unaligned base): the
    // consumers fill a double-buffered box with 4-byte cp.async copies
    // (out-of-grid cells are zero, as TMA's fill) while computing the other
    static_assert(S == 2, "LDG variant double-buffers");
    static_assert(BX % 2 == 0 && XH % 2 == 0 && TX % 2 == 0 && C::BOX_FLOATS % 2 == 0, "pair fill");
    // even nx and 8-B aligned bases (e.g. SHOC's 4098-wide rows): the box is
    // filled in 8-byte pairs; x0 - XH is even, so a pair is wholly in or out
    const bool pairs = (nx % 2 == 0) && ((reinterpret_cast<uintptr_t>(src0) | reinterpret_cast<uintptr_t>(src1)) & 7u) == 0;
    auto fill = [&](int s, int64_t t) {
      const int x0 = (int)(t % ntx) * TX, y0 = (int)(t / ntx) * TY;
      float* base = reinterpret_cast<float*>(dsm4 + s * SF4);
      if (pairs) {
        constexpr int BX2 = BX / 2;
        for (int idx = threadIdx.x; idx < NIN * C::BY * BX2; idx += NCONS) {
          const int b = idx / (C::BY * BX2), rem = idx % (C::BY * BX2);
          const int r = rem / BX2, c = 2 * (rem % BX2);
          const int gy = y0 - RY + r, gx = x0 - XH + c;
          float* dst = base + b * C::BOX_FLOATS + r * BX + c;
          if (gy >= 0 && gy < ny && gx >= 0 && gx < nx)
            cp_async8(dst, (b == 0 ? src0 : src1) + (int64_t)gy * nx + gx);
          else
            *reinterpret_cast<float2*>(dst) = make_float2(0.0f, 0.0f);
        }
        cp_async_commit();
        return;
      }
      for (int idx = threadIdx.x; idx < NIN * C::BY * BX; idx += NCONS) {
        const int b = idx / (C::BY * BX), rem = idx % (C::BY * BX);
        const int r = rem / BX, c = rem % BX;
        const int gy = y0 - RY + r, gx = x0 - XH + c;
        float* dst = base + b * C::BOX_FLOATS + r * BX + c;
        if (gy >= 0 && gy < ny && gx >= 0 && gx < nx)
          cp_async4(dst, (b == 0 ? src0 : src1) + (int64_t)gy * nx + gx);
        else
          *dst = 0.0f;
      }
      cp_async_commit();
    };
    fill(0, blockIdx.x);
    for (int i = 0; i < nt; ++i) {
      const int64_t t = blockIdx.x + (int64_t)i * gridDim.x;
      if (i + 1 < nt) {
        fill((i + 1) & 1, t + gridDim.x);
        cp_async_wait<1>();
      } else {
        cp_async_wait<0>();
      }
      named_bar_sync(1, NCONS);
      const int x0 = (int)(t % ntx) * TX, y0 = (int)(t / ntx) * TY;
      fixup(i & 1, x0, y0);
      compute(i & 1, x0, y0);
      named_bar_sync(1, NCONS);       // the next fill reuses this stage
    }
  }
}

// ---------------------------------------------------------------------------
// K1S: one full SRAD iteration fused into one tile pass:
// I' = SRAD2(c, I) with c = SRAD1(I) computed on the fly for the tile's rows
// plus one row below and one column to the right (the S and E taps of
// SRAD2), never stored.  The I box is (128+8) x (TY+4) at (x0-4, y0-2); each
// warp keeps 4 I x-windows and 3 c rows in registers while sweeping its rows.
// c is a grid read through the same pad as I: out-of-grid c rows/columns
// take the value at the remapped position.  Every value goes through
// op_srad1 / op_srad2, so the result equals SRAD1 then SRAD2 bit for bit.
// ---------------------------------------------------------------------------
template <int RX, int I>
struct RowsAcc {                 // rows[0..2] = I rows y-1, y, y+1 (x-windows with offsets -RX..)
  const float* r0;
  const float* r1;
  const float* r2;
  template <int DZ, int DY, int DX>
  __device__ __forceinline__ float at() const {
    static_assert(DZ == 0, "2D");
    return DY < 0 ? r0[I + RX + DX] : (DY > 0 ? r2[I + RX + DX] : r1[I + RX + DX]);
  }
};

template <int I>
struct CRowsAcc {                // c at (y, x+i) = cy[i], (y+1, x+i) = cs[i]
  const float* cy;
  const float* cs;
  template <int DZ, int DY, int DX>
  __device__ __forceinline__ float at() const {
    static_assert(DZ == 0 && DY >= 0 && DX >= 0, "SRAD2 reads c at C, S, E");
    return DY > 0 ? cs[I + DX] : cy[I + DX];
  }
};

template <int RPW, int S, int MINB>
__global__ void __launch_bounds__(NCONS + 32, MINB)
    k1_srad_fused(const __grid_constant__ StencilParams p, const __grid_constant__ CUtensorMap map0,
                  const float* __restrict__ src0, float* __restrict__ out, int ntx, int nty) {
  using C = Cfg<2, RPW, S, 1>;
  constexpr int TY = C::TY;
  constexpr int W = 8;            // x-window offsets -2 .. +5
  constexpr int BX4 = BX / 4;
  constexpr int SF4 = C::STAGE_FLOATS / 4;
  extern __shared__ __align__(128) float4 dsm4[];
  uint64_t* full = reinterpret_cast<uint64_t*>(dsm4 + S * SF4);
  uint64_t* empty = full + S;
  const int64_t ntiles = (int64_t)ntx * nty;
  const int nt = (int)((ntiles - blockIdx.x + gridDim.x - 1) / gridDim.x);
  if (nt <= 0) return;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  if (threadIdx.x == 0) {
    for (int s = 0; s < S; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NW);
    }
    fence_mbar_init();
  }
  __syncthreads();
  pdl_launch_dependents();   // PDL: let the next launch ramp up now
  pdl_wait();                // ... and wait for the previous one before any global access
  if (warp == NW) {
    if (lane == 0) {
      prefetch_tmap(&map0);
      int s = 0;
      uint32_t pass = 0;
      for (int i = 0; i < nt; ++i) {
        if (pass > 0) mbar_wait(&empty[s], (pass - 1) & 1);
        const int64_t t = blockIdx.x + (int64_t)i * gridDim.x;
        const int x0 = (int)(t % ntx) * TX, y0 = (int)(t / ntx) * TY;
        mbar_arrive_expect_tx(&full[s], C::BOX_BYTES);
        tma_load_3d(dsm4 + s * SF4, &map0, &full[s], x0 - XH, y0 - 2, 0);
        if (++s == S) { s = 0; ++pass; }
      }
    }
    return;
  }
  const int nx = (int)p.n[2], ny = (int)p.n[1];
  const int kx = p.kind[2], ky = p.kind[1];
  // q0 of the input image: reduce the previous pass's (or k_sum2's) fp64
  // partials here, in a fixed order (so every CTA gets the same bits), while
  // the producer's first TMA loads are already in flight
  __shared__ double2 s_red[NW];
  float q[3];                      // SRAD1's constants {q0, a, b} in registers
  if (!p.srad_part_in) {
#pragma unroll
    for (int k = 0; k < 3; ++k) q[k] = p.srad_q0[k];
  } else {
    constexpr int K = kSradMaxParts / NCONS;
    double2 v[K];
#pragma unroll
    for (int k = 0; k < K; ++k) {
      const int i = threadIdx.x + k * NCONS;
      v[k] = i < p.srad_nparts ? p.srad_part_in[i] : make_double2(0.0, 0.0);
    }
    double a = 0.0, b = 0.0;
#pragma unroll
    for (int k = 0; k < K; ++k) {
      a += v[k].x;
      b += v[k].y;
    }
    for (int o = 16; o > 0; o >>= 1) {
      a += __shfl_down_sync(0xffffffffu, a, o);
      b += __shfl_down_sync(0xffffffffu, b, o);
    }
    if (lane == 0) s_red[warp] = make_double2(a, b);
    named_bar_sync(1, NCONS);
    a = b = 0.0;
#pragma unroll
    for (int w = 0; w < NW; ++w) {
      a += s_red[w].x;
      b += s_red[w].y;
    }
    srad1_constants(srad_q0sqr(a, b, p.n[1] * p.n[2]), q);
    named_bar_sync(1, NCONS);      // s_red is reused for this pass's own statistics
  }
  double st_s = 0.0, st_ss = 0.0;  // statistics of the written image (next iteration's q0)
  const int r0 = warp * RPW;
  int s = 0;
  uint32_t pass = 0;
  for (int it = 0; it < nt; ++it) {
    mbar_wait(&full[s], pass & 1);
    const int64_t t = blockIdx.x + (int64_t)it * gridDim.x;
    const int x0 = (int)(t % ntx) * TX, y0 = (int)(t / ntx) * TY;
    const bool edge = (x0 == 0) || (x0 + TX + 2 > nx) || (y0 < 2) || (y0 + TY + 2 > ny);
    if (edge) {
      // every warp is past this stage's previous tile (guaranteed already by
      // the empty/full mbarrier hand-off; the barrier makes it explicit to
      // racecheck, edge tiles only)
      named_bar_sync(1, NCONS);
      fixup_tile<2, 2, XH, BX, C::BY, NCONS>(p, reinterpret_cast<float*>(dsm4 + s * SF4), src0, 0, x0, y0,
                                             threadIdx.x);
      fence_proxy_async_smem();
      named_bar_sync(1, NCONS);
    }
    const int xo = x0 + 4 * lane;
    const bool x_ok = xo < nx;
    // c column x+4 at the right grid edge takes the remapped column's value;
    // under WRAP the fixed-up box already holds I's wrapped columns, so the
    // value SRAD1 computes there IS c(0) (the remap would point at
    // column -xo)
    const int ce = (xo + 4 == nx && kx != PAD_WRAP) ? (int)(pad_remap(nx, nx, kx) - xo) : 4;
    const float4* box = dsm4 + s * SF4;
    float iw[4][W];
    float cr[3][5];
    float* orow = out + ((int64_t)(y0 + r0) * nx + xo);
    // c at the tile's right halo column x0 + 128 (SRAD2's E tap of lane 31)
    // for this warp's RPW + 1 c rows, one row per lane (lanes 0..RPW): every
    // other lane's column x + 4 is its right neighbour's column x (shuffle),
    // so each lane evaluates SRAD1 for 4 columns instead of 5
    float halo_c;
    {
      const int j = lane < RPW + 1 ? lane : RPW;
      const float* bf = reinterpret_cast<const float*>(box) + (r0 + j + 1) * BX + TX + XH - 1;
      float a0[3], a1[3], a2[3];
#pragma unroll
      for (int d = 0; d < 3; ++d) {
        a0[d] = bf[d];
        a1[d] = bf[BX + d];
        a2[d] = bf[2 * BX + d];
      }
      halo_c = op_srad1(RowsAcc<1, 0>{a0, a1, a2}, q);
    }
    // box rows r0+1 .. r0+RPW+3  <->  I rows y0+r0-1 .. y0+r0+RPW+1
    static_for<RPW + 3>([&](auto K) {
      constexpr int k = decltype(K)::value;
      load_row<2>(box + (r0 + 1 + k) * BX4, lane, iw[k % 4]);
      if constexpr (k >= 2) {
        // c for I row crow = y0 + r0 + k - 2 from I rows crow-1 .. crow+1
        constexpr int cs_ = (k - 2) % 3;
        const int crow = y0 + r0 + k - 2;
        // c rows past the bottom edge: WRAP computes them from the box's
        // wrapped I rows (= c(crow - ny)); the others copy the remapped row
        if (crow < ny || ky == PAD_WRAP) {
          static_for<4>([&](auto II) {
            constexpr int ii = decltype(II)::value;
            cr[cs_][ii] = op_srad1(RowsAcc<2, ii>{iw[(k - 2) % 4], iw[(k - 1) % 4], iw[k % 4]}, q);
          });
          const float right = __shfl_down_sync(0xffffffffu, cr[cs_][0], 1);
          const float hcol = __shfl_sync(0xffffffffu, halo_c, k - 2);
          float e4 = lane == 31 ? hcol : right;
          if (ce != 4) e4 = ce == 3 ? cr[cs_][3] : (ce == 2 ? cr[cs_][2] : cr[cs_][1]);   // the grid's last column
          cr[cs_][4] = e4;
        } else if constexpr (k >= 3) {
          // c row outside the grid: the remapped row (one or two above)
          const int d = crow - (int)pad_remap(crow, ny, ky);
#pragma unroll
          for (int ii = 0; ii < 5; ++ii) {
            if constexpr (k >= 4)
              cr[cs_][ii] = d == 1 ? cr[(k - 3) % 3][ii] : cr[(k - 4) % 3][ii];
            else
              cr[cs_][ii] = cr[(k - 3) % 3][ii];
          }
        }
      }
      if constexpr (k >= 3) {
        // output row o = k - 3 (I row y0 + r0 + o)
        constexpr int o = k - 3;
        if constexpr (o < RPW) {
          float v[4];
          static_for<4>([&](auto II) {
            constexpr int ii = decltype(II)::value;
            v[ii] = op_srad2(CRowsAcc<ii>{cr[o % 3], cr[(o + 1) % 3]},
                             RowsAcc<2, ii>{iw[o % 4], iw[(o + 1) % 4], iw[(o + 2) % 4]}, p.prm);
          });
          if (x_ok && y0 + r0 + o < ny) {
            stg128(orow + (int64_t)o * nx, make_float4(v[0], v[1], v[2], v[3]));
#pragma unroll
            for (int ii = 0; ii < 4; ++ii) {
              const double d = v[ii];
              st_s += d;
              st_ss = fma(d, d, st_ss);
            }
          }
        }
      }
    });
    __syncwarp();
    if (lane == 0) mbar_arrive(&empty[s]);
    if (++s == S) { s = 0; ++pass; }
  }
  if (p.srad_part_out) {
    for (int o = 16; o > 0; o >>= 1) {
      st_s += __shfl_down_sync(0xffffffffu, st_s, o);
      st_ss += __shfl_down_sync(0xffffffffu, st_ss, o);
    }
    if (lane == 0) s_red[warp] = make_double2(st_s, st_ss);
    named_bar_sync(1, NCONS);
    if (threadIdx.x == 0) {
      double a = 0.0, b = 0.0;
      for (int w = 0; w < NW; ++w) {
        a += s_red[w].x;
        b += s_red[w].y;
      }
      p.srad_part_out[blockIdx.x] = make_double2(a, b);
    }
  }
}

struct Launcher {
  const void* fn;
  int smem;
  int ty;
  int ry;
  int nin;
  int ctas_per_sm;
};

template <int OP, int RY, int RX, int RPW, int S, int NIN, int MINB = 3, bool LDG = false>
Launcher get_launcher() {
  static Launcher L{};
  static std::once_flag once;
  std::call_once(once, [] {
    using C = Cfg<RY, RPW, S, NIN>;
    auto fn = k1_tile<OP, RY, RX, RPW, S, NIN, MINB, LDG>;
    cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, C::SMEM);
    int occ = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, fn, NCONS + 32, C::SMEM) != cudaSuccess) occ = 1;
    cudaGetLastError();
    L = Launcher{reinterpret_cast<const void*>(fn), C::SMEM, C::TY, RY, NIN, occ > 0 ? occ : 1};
  });
  return L;
}

bool star2d(const StencilParams& p, int RY, int RX) {
  const int SX = 2 * RX + 1;
  for (int ky = 0; ky < 2 * RY + 1; ++ky)
    for (int kx = 0; kx < SX; ++kx)
      if (ky != RY && kx != RX && p.wbox[ky * SX + kx] != 0.0f) return false;
  return true;
}

// Tile shape per launch: small grids (fewer 128 x 48 tiles than SMs, e.g.
// J2D5 256^2, SRAD 504x458) take 128 x 8 tiles (6x the CTAs, each a sixth
// of the latency chain); otherwise (rows per warp, stages, CTAs per SM) =
// (4, 4, 2) for the separable Gaussian — a 4-deep ring of 128 x 32 tiles
// keeps more bytes in flight — and (6, 2, 3) for SRAD (measured per op,
// profiles/r01_sweep_k1_shapes_k3.txt); LIFT_K1_SHAPE overrides
// (1 = (6, 2, 3), 2 = (4, 3, 3), 3 = (8, 3, 2), 4 = (4, 4, 2))
template <int OPV, int RYV, int RXV, int NINV>
Launcher pick_k1(bool ldg, bool small) {
  if (ldg) return get_launcher<OPV, RYV, RXV, 6, 2, NINV, 3, true>();
  if (small) return get_launcher<OPV, RYV, RXV, 1, 2, NINV, 4, false>();
  const char* e = getenv("LIFT_K1_SHAPE");
  switch (e ? atoi(e) : (OPV == K1_WSEP ? 4 : 1)) {
    case 2: return get_launcher<OPV, RYV, RXV, 4, 3, NINV, 3, false>();
    case 3: return get_launcher<OPV, RYV, RXV, 8, 3, NINV, 2, false>();
    case 4: return get_launcher<OPV, RYV, RXV, 4, 4, NINV, 2, false>();
    default: return get_launcher<OPV, RYV, RXV, 6, 2, NINV, 3, false>();
  }
}
#define K1_PICK(OPV, RYV, RXV, NINV) pick_k1<OPV, RYV, RXV, NINV>(ldg, small)

bool pick(const StencilParams& p, bool ldg, bool small, Launcher* L) {
  const int ry = p.lo[1], rx = p.lo[2];
  if (p.op == OP_WEIGHTED) {
    const int mode = p.sep ? K1_WSEP : (star2d(p, ry, rx) ? K1_WSTAR : K1_WBOX);
#define K1_CASE(RYV, RXV)                                                     \
  if (ry == RYV && rx == RXV) {                                              \
    if (mode == K1_WSEP) *L = K1_PICK(K1_WSEP, RYV, RXV, 1);                 \
    else if (mode == K1_WSTAR) *L = K1_PICK(K1_WSTAR, RYV, RXV, 1);          \
    else *L = K1_PICK(K1_WBOX, RYV, RXV, 1);                                 \
    return true;                                                             \
  }
    K1_CASE(1, 1)
    K1_CASE(2, 2)
    K1_CASE(1, 2)
    K1_CASE(2, 1)
#undef K1_CASE
    return false;
  }
  if (p.op == OP_SRAD1) { *L = K1_PICK(K1_SRAD1, 1, 1, 1); return true; }
  if (p.op == OP_SRAD2) { *L = K1_PICK(K1_SRAD2, 1, 1, 2); return true; }
  if (p.op == OP_HOTSPOT2D) { *L = K1_PICK(K1_HOT2D, 1, 1, 2); return true; }
  if (p.op == OP_GRADIENT) { *L = K1_PICK(K1_GRAD, 1, 1, 1); return true; }
  return false;
}

struct MapEntry {
  const float* base;
  int64_t nx, ny;
  int by;
  CUtensorMap map;
};

bool get_map(const float* base, int64_t nx, int64_t ny, int by, CUtensorMap* out, std::string* err) {
  thread_local MapEntry cache[8];
  thread_local int next = 0;
  for (auto& e : cache)
    if (e.base == base && e.nx == nx && e.ny == ny && e.by == by) {
      *out = e.map;
      return true;
    }
  MapEntry e{base, nx, ny, by, {}};
  if (!encode_tensor_map_3d(&e.map, base, nx, ny, 1, BX, (uint32_t)by, 1, err)) return false;
  cache[next] = e;
  next = (next + 1) % 8;
  *out = e.map;
  return true;
}

}  // namespace

template <int RPW, int S, int MINB>
Launcher srad_fused_launcher() {
  static Launcher L{};
  static std::once_flag once;
  std::call_once(once, [] {
    using C = Cfg<2, RPW, S, 1>;
    auto fn = k1_srad_fused<RPW, S, MINB>;
    cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, C::SMEM);
    int occ = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, fn, NCONS + 32, C::SMEM) != cudaSuccess) occ = 1;
    cudaGetLastError();
    L = Launcher{reinterpret_cast<const void*>(fn), C::SMEM, C::TY, 2, 1, occ > 0 ? occ : 1};
  });
  return L;
}

cudaError_t launch_srad_fused(const StencilParams& p, const float* in0, float* out, cudaStream_t stream,
                              int num_sms, std::string* err, int* nparts_out) {
  // (rows per warp, stages, min CTAs/SM); LIFT_SRAD_SHAPE overrides (A/B sweeps)
  const char* env = getenv("LIFT_SRAD_SHAPE");
  Launcher L;
  switch (env ? atoi(env) : 0) {
    case 1: L = srad_fused_launcher<6, 2, 2>(); break;
    case 2: L = srad_fused_launcher<4, 3, 2>(); break;
    case 3: L = srad_fused_launcher<6, 3, 2>(); break;
    case 4: L = srad_fused_launcher<4, 2, 3>(); break;
    case 5: L = srad_fused_launcher<8, 2, 3>(); break;
    case 6: L = srad_fused_launcher<6, 2, 3>(); break;     // round 1's default
    case 7: L = srad_fused_launcher<12, 2, 2>(); break;
    // 8 rows per warp (SRAD1 for 9/8 instead of 7/6 of the rows), 96
    // registers without spills at 2 CTAs/SM: 379 -> 386 Gpts/s
    // (profiles/r02_ab_srad_shape.txt)
    default: L = srad_fused_launcher<8, 2, 2>(); break;
  }
  CUtensorMap m0;
  if (!get_map(in0, p.n[2], p.n[1], L.ty + 4, &m0, err)) return cudaErrorInvalidValue;
  const int ntx = (int)((p.n[2] + TX - 1) / TX);
  const int nty = (int)((p.n[1] + L.ty - 1) / L.ty);
  int64_t grid = (int64_t)num_sms * L.ctas_per_sm;
  if (grid > (int64_t)ntx * nty) grid = (int64_t)ntx * nty;
  if (p.srad_part_in && p.srad_nparts > kSradMaxParts) {
    *err = "SRAD: too many q0 partials";
    return cudaErrorInvalidValue;
  }
  if (nparts_out) *nparts_out = (int)grid;
  void* args[] = {(void*)&p, (void*)&m0, (void*)&in0, (void*)&out, (void*)&ntx, (void*)&nty};
  set_last_kernel("k1_srad_fused");
  return launch_kernel(L.fn, dim3((unsigned)grid), dim3(NCONS + 32), args, (size_t)L.smem, stream, true);
}

bool tile2d_supported(const StencilParams& p) {
  if (has_dampen(p)) return false;     // DAMPEN pads run on K5 / K0
  // canonical 2D plan: dimension 0 is the dummy (extent 1, size 1, no pad)
  if (p.n[0] != 1 || p.size[0] != 1 || p.lo[0] != 0 || p.hi[0] != 0 || p.slab) return false;
  const int ry = p.lo[1], rx = p.lo[2];
  for (int d = 1; d < 3; ++d)
    if (p.step[d] != 1 || p.hi[d] != p.lo[d] || p.size[d] != 2 * p.lo[d] + 1) return false;
  if (ry < 1 || ry > 2 || rx < 1 || rx > 2) return false;
  if (p.op == OP_SRAD1 || p.op == OP_SRAD2 || p.op == OP_HOTSPOT2D || p.op == OP_GRADIENT || p.op == OP_SRAD) {
    if (ry != 1 || rx != 1) return false;
  } else if (p.op != OP_WEIGHTED) {
    return false;
  }
  if (p.op == OP_SRAD && p.n[2] % 4 != 0) return false;   // the fused SRAD pass is TMA-only
  if (p.n[2] * p.n[1] >= (1ll << 31)) return false;
  return true;
}

cudaError_t launch_tile2d(const StencilParams& p, const float* in0, const float* in1, float* out,
                          cudaStream_t stream, int num_sms, std::string* err) {
  if (p.op == OP_SRAD) return launch_srad_fused(p, in0, out, stream, num_sms, err, nullptr);
  const bool small = ((p.n[2] + TX - 1) / TX) * ((p.n[1] + 6 * NW - 1) / (6 * NW)) < num_sms;
  // per-warp streaming sweeps (K3) where they measured faster than the tiles
  if (wsweep2d_supported(p, in0, in1, small)) return launch_wsweep2d(p, in0, in1, out, stream, num_sms, err);
  // TMA needs 16-B aligned bases and row pitches; otherwise cp.async fills the box
  const bool ldg = (p.n[2] % 4 != 0) || (reinterpret_cast<uintptr_t>(in0) & 15u) ||
                   (in1 && (reinterpret_cast<uintptr_t>(in1) & 15u));
  Launcher L;
  if (!pick(p, ldg, small, &L)) {
    *err = "tile2d: no instantiation";
    return cudaErrorNotSupported;
  }
  CUtensorMap m0{}, m1{};
  if (!ldg) {
    if (!get_map(in0, p.n[2], p.n[1], L.ty + 2 * L.ry, &m0, err)) return cudaErrorInvalidValue;
    if (L.nin > 1) {
      if (!get_map(in1, p.n[2], p.n[1], L.ty + 2 * L.ry, &m1, err)) return cudaErrorInvalidValue;
    } else {
      m1 = m0;
    }
  }
  const int ntx = (int)((p.n[2] + TX - 1) / TX);
  const int nty = (int)((p.n[1] + L.ty - 1) / L.ty);
  const int64_t ntiles = (int64_t)ntx * nty;
  int64_t grid = (int64_t)num_sms * L.ctas_per_sm;
  if (grid > ntiles) grid = ntiles;
  const float* s1 = L.nin > 1 ? in1 : in0;
  void* args[] = {(void*)&p, (void*)&m0, (void*)&m1, (void*)&in0, (void*)&s1, (void*)&out, (void*)&ntx, (void*)&nty};
  set_last_kernel("k1_tile");
  return launch_kernel(L.fn, dim3((unsigned)grid), dim3(NCONS + 32), args, (size_t)L.smem, stream, true);
}

}  // namespace lift
