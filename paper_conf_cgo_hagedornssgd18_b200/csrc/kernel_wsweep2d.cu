// kernel_wsweep2d.cu — K3: the 2D stencil as independent per-warp y-sweeps.
//
// map_2(f, slide_2(size, step, pad_2(...))) over a 2D
// grid, with the overlapped tiling of P:693-822 cut the other way round from
// K1: a work item is a 128-column strip of a chunk of rows, and ONE warp owns
// it from top to bottom.  Each warp is its own TMA pipeline: lane 0 keeps S
// groups of G input rows ((128+8) x G floats per input grid, one tensor-map
// box) in flight in the warp's private shared-memory ring and refills a slot
// as soon as the warp has consumed it — no producer warp, no CTA barrier, no
// empty barriers.  Items come from a global ticket counter, and the load
// cursor runs into the next item while the current one is consumed, so a
// warp never drains its pipeline between items.  Every input row is read from
// shared memory once (one LDS.128 per lane, in-row neighbours by shuffles)
// and added to the 2RY+1 output rows in flight (weighted ops; the same
// row-major tap order as K0/K1, so results are bitwise identical), or kept in
// a ring of 2RY+1 x-windows (SRAD, Hotspot2D, Gradient).
//
// pad: every group is one box load (rows outside the grid are TMA's zero
// fill).  Items whose chunk or strip touches the grid boundary run a general
// copy of the sweep: a row outside [0, ny) is read from its remapped row in
// global memory (L2) for CLAMP / MIRROR / REFLECT / WRAP, or is the pad value
// for CONSTANT; x taps outside [0, nx) are selected from the lane's own float4
// (CLAMP / MIRROR / REFLECT, R <= 2 < 4) or are the pad value.  Interior items
// run a copy without any of this.  WRAP in x and untileable rows (nx % 4 !=
// 0, unaligned bases) run on K1.
#include <cuda.h>
#include <cuda_runtime.h>

#include <algorithm>
#include <atomic>
#include <cstdlib>
#include <mutex>
#include <string>

#include "common.cuh"
#include "launch.hpp"
#include "ops.cuh"
#include "slots.cuh"
#include "tma.cuh"

namespace lift {
namespace {

constexpr int TX = 128;
constexpr int XH = 4;
constexpr int BX = TX + 2 * XH;
constexpr int BX4 = BX / 4;
constexpr unsigned FULL = 0xffffffffu;
// dynamic work counters, one slot per running launch (slots.cuh): c[0] item
// ticket, c[1] CTAs done
__device__ LaunchSlot g_launch[kLaunchSlots];

enum K3Op { K3_WBOX = 0, K3_SRAD1 = 1, K3_SRAD2 = 2, K3_WSTAR = 3, K3_WSEP = 4, K3_HOT2D = 5, K3_GRAD = 6 };

template <int G, int S, int NIN, int WPC>
struct WCfg {
  static_assert(G % 4 == 0, "G rows of 544 B keep every box 128-B aligned");
  static_assert((G & (G - 1)) == 0, "row-in-group is i & (G - 1)");
  static constexpr int GROUP_FLOATS = BX * G;            // one input grid, one group
  static constexpr int SLOT_FLOATS = NIN * GROUP_FLOATS;
  static constexpr int WARP_FLOATS = S * SLOT_FLOATS;
  static constexpr int SMEM = WPC * (WARP_FLOATS * 4 + S * 8) + 128;
};

// out-of-grid x tap selection for the lane's 4 outputs: -2 keep, -1 the pad
// value, 0..3 the element of the lane's own float4
template <int RX>
struct XSel {
  int l[RX > 0 ? RX : 1];
  int r[RX > 0 ? RX : 1];
};

__device__ __forceinline__ float sel4(int s, const float (&c)[4], float pv) {
  return s < 0 ? pv : (s == 0 ? c[0] : (s == 1 ? c[1] : (s == 2 ? c[2] : c[3])));
}

// x-window of one row for the 4 outputs of a lane (offsets -RX .. 3+RX)
// from the lane's float4 c and its row's halo float4 e (left one for lane 0,
// right one for lane 31)
template <int RX, bool XE>
__device__ __forceinline__ void make_window(const float4 c, const float4 e, int lane, float (&xw)[4 + 2 * RX],
                                            const XSel<RX>& xs, float pv) {
  const float cv[4] = {c.x, c.y, c.z, c.w};
  const float ev[4] = {e.x, e.y, e.z, e.w};
#pragma unroll
  for (int k = 1; k <= RX; ++k) {
    float l = __shfl_up_sync(FULL, cv[4 - k], 1);     // x - k from the left lane
    float r = __shfl_down_sync(FULL, cv[k - 1], 1);   // x + 3 + k from the right lane
    if (lane == 0) l = ev[4 - k];
    if (lane == 31) r = ev[k - 1];
    if constexpr (XE) {
      if (xs.l[k - 1] > -2) l = sel4(xs.l[k - 1], cv, pv);
      if (xs.r[k - 1] > -2) r = sel4(xs.r[k - 1], cv, pv);
    }
    xw[RX - k] = l;
    xw[RX + 3 + k] = r;
  }
#pragma unroll
  for (int i = 0; i < 4; ++i) xw[RX + i] = cv[i];
}

// the same from a staged box row in shared memory
template <int RX, bool XE>
__device__ __forceinline__ void load_row(const float4* row4, int lane, float (&xw)[4 + 2 * RX], const XSel<RX>& xs,
                                         float pv) {
  make_window<RX, XE>(row4[XH / 4 + lane], row4[lane == 0 ? 0 : (TX + XH) / 4], lane, xw, xs, pv);
}

// the lane's float4 and halo float4 of a staged row (shared memory) or, for
// a remapped out-of-grid row of an edge item, of grid row y in global memory;
// no shuffles here, so the (warp-uniform) choice stays outside collective code
template <bool XE>
__device__ __forceinline__ void fetch_row(const float4* row4, const float* __restrict__ src, int y, int x0, int nx,
                                          int lane, float4& c, float4& e) {
  if (XE && y >= 0) {
    const float* row = src + (int64_t)y * nx;
    const int xo = x0 + 4 * lane;
    const float4 z = make_float4(0.f, 0.f, 0.f, 0.f);
    c = xo < nx ? ldg128(row + xo) : z;
    const int xe = lane == 0 ? x0 - XH : x0 + TX;
    e = (xe >= 0 && xe < nx) ? ldg128(row + xe) : z;
  } else {
    c = row4[XH / 4 + lane];
    e = row4[lane == 0 ? 0 : (TX + XH) / 4];
  }
}

template <int RY, int RX, int I>
struct RingAcc {
  const float (*rows)[4 + 2 * RX];
  template <int DZ, int DY, int DX>
  __device__ __forceinline__ float at() const {
    static_assert(DZ == 0, "2D");
    return rows[DY + RY][I + RX + DX];
  }
};

struct Item {
  int x0, y0, nout, nin, ng;   // strip origin, output rows, input rows, groups
};

template <int OP, int RY, int RX, int G, int S, int NIN, int WPC, int MINB>
__global__ void __launch_bounds__(WPC * 32, MINB)
    k3_wsweep(const __grid_constant__ StencilParams p, const __grid_constant__ CUtensorMap map0,
              const __grid_constant__ CUtensorMap map1, const float* __restrict__ src0,
              const float* __restrict__ src1, float* __restrict__ out, int nstrips, int hc, int nitems) {
  using C = WCfg<G, S, NIN, WPC>;
  constexpr int SY = 2 * RY + 1, SX = 2 * RX + 1;
  constexpr int W = 4 + 2 * RX;
  // accumulator / window ring: RS >= SY slots, a multiple of G, so the slot
  // of row i (i mod RS) is compile-time within a block of U = RS / G groups
  constexpr int RS = ((SY + G - 1) / G) * G;
  constexpr int U = RS / G;
  constexpr bool WEIGHTED = OP == K3_WBOX || OP == K3_WSTAR || OP == K3_WSEP;
  constexpr int SLOT4 = C::SLOT_FLOATS / 4;
  constexpr int GROUP4 = C::GROUP_FLOATS / 4;
  constexpr uint32_t TXB = NIN * G * BX * 4;   // bytes per slot

  extern __shared__ __align__(128) float4 dsm4[];
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  float4* ring = dsm4 + warp * (S * SLOT4);
  uint64_t* bars = reinterpret_cast<uint64_t*>(dsm4 + WPC * (S * SLOT4)) + warp * S;

  int slot = 0;
  if (lane == 0) {
    for (int s = 0; s < S; ++s) mbar_init(&bars[s], 1);
    fence_mbar_init();
    prefetch_tmap(&map0);
    if constexpr (NIN > 1) prefetch_tmap(&map1);
    slot = claim_launch_slot(g_launch);    // the same slot in every warp of the launch
  }
  slot = __shfl_sync(FULL, slot, 0);
  __syncwarp();
  pdl_launch_dependents();
  pdl_wait();

  const int nx = (int)p.n[2], ny = (int)p.n[1];
  const int kx = p.kind[2], ky = p.kind[1];
  const float pv = p.pad_value;
  const bool kyc = ky == PAD_CONSTANT;
  const bool kyc_nz = kyc && pv != 0.0f;     // constant rows that TMA's zero fill does not give
  const bool vec = (reinterpret_cast<uintptr_t>(out) & 15u) == 0;

  auto geo = [&](int item) {
    Item it;
    const int s = item % nstrips, c = item / nstrips;
    it.x0 = s * TX;
    it.y0 = c * hc;
    it.nout = min(hc, ny - it.y0);
    it.nin = it.nout + 2 * RY;
    it.ng = ((it.nin + RS - 1) / RS) * U;   // whole blocks (the tail rows are computed, not stored)
    return it;
  };
  auto fetch = [&]() {
    int v = 0;
    if (lane == 0) v = (int)atomicAdd(&g_launch[slot].c[0], 1u);
    return __shfl_sync(FULL, v, 0);
  };

  // ---- load cursor (lane 0 issues; every lane tracks it identically)
  int l_item = fetch();
  Item lg = geo(l_item < nitems ? l_item : 0);
  int l_g = 0;
  int ls = 0;             // next slot to fill
  int inflight = 0;
  int c_item = l_item;    // item being consumed
  auto issue = [&]() {
    if (lane == 0) {
      uint64_t* bar = &bars[ls];
      float* dst = reinterpret_cast<float*>(ring + ls * SLOT4);
      const int yb = lg.y0 - RY + l_g * G;
      mbar_arrive_expect_tx(bar, TXB);
      tma_load_3d(dst, &map0, bar, lg.x0 - XH, yb, 0);
      if constexpr (NIN > 1) tma_load_3d(dst + C::GROUP_FLOATS, &map1, bar, lg.x0 - XH, yb, 0);
    }
    if (++ls == S) ls = 0;
    ++l_g;
    ++inflight;
  };
  // keep S groups in flight, running at most one item ahead of the consumer
  auto refill = [&]() {
    while (inflight < S && l_item < nitems) {
      if (l_g == lg.ng) {
        if (l_item != c_item) break;        // already one item ahead
        l_item = fetch();
        if (l_item >= nitems) break;
        lg = geo(l_item);
        l_g = 0;
      }
      issue();
    }
  };
  refill();

  int cs = 0;             // next slot to consume
  uint32_t cphase = 0;    // parity bits per slot
  while (c_item < nitems) {
    const Item it = geo(c_item);
    const int xo = it.x0 + 4 * lane;
    const bool x_ok = xo < nx;
    // general (edge) sweep: the strip touches the x boundary, or the chunk's
    // halo rows leave the grid
    const bool edge = (it.x0 == 0) || (it.x0 + TX + RX > nx) || (it.y0 < RY) || (it.y0 + it.nout + RY > ny);
    XSel<RX> xs;
#pragma unroll
    for (int k = 1; k <= RX; ++k) {
      xs.l[k - 1] = -2;
      xs.r[k - 1] = -2;
      if (xo - k < 0) xs.l[k - 1] = kx == PAD_CONSTANT ? -1 : (int)pad_remap(xo - k, nx, kx) - xo;
      if (xo < nx && xo + 3 + k >= nx)
        xs.r[k - 1] = kx == PAD_CONSTANT ? -1 : (int)pad_remap(xo + 3 + k, nx, kx) - xo;
    }
    float* obase = out + (int64_t)it.y0 * nx + xo;

    auto sweep = [&](auto XE_) {
      constexpr bool XE = decltype(XE_)::value;
      float acc[WEIGHTED ? RS : 1][4];
      float ra[WEIGHTED ? 1 : RS][W];
      float rb[(!WEIGHTED && NIN > 1) ? RS : 1][W];
      auto store = [&](int o, const float (&v)[4]) {
        if (!(x_ok && o >= 0 && o < it.nout)) return;
        float* dst = obase + (int64_t)o * nx;
        if (vec) {
          stg128(dst, make_float4(v[0], v[1], v[2], v[3]));
        } else {
#pragma unroll
          for (int q = 0; q < 4; ++q) dst[q] = v[q];
        }
      };
      // one input row i (chunk-relative; input row y0 - RY + i); R = i mod (SY*G) is compile-time
      auto row = [&](auto R_, int i, const float4* row0, const float4* row1) {
        constexpr int R = decltype(R_)::value;
        constexpr int rs = R % RS;
        float xw[W];
        // rows outside the grid (general sweep only): CONSTANT -> the value
        // (TMA's zero fill when it is 0), otherwise the remapped row h_y(y)
        // from global memory
        int yrow = -1;
        bool yconst = false;
        if constexpr (XE) {
          const int y = it.y0 - RY + i;
          if (y < 0 || y >= ny) {
            if (kyc) yconst = kyc_nz;
            else yrow = (int)pad_remap(y, ny, ky);
          }
        }
        {
          float4 c, e;
          fetch_row<XE>(row0, src0, yrow, it.x0, nx, lane, c, e);
          make_window<RX, XE>(c, e, lane, xw, xs, pv);
        }
        if (XE && yconst) {
#pragma unroll
          for (int q = 0; q < W; ++q) xw[q] = pv;
        }
        if constexpr (WEIGHTED) {
          float h[4];
          if constexpr (OP == K3_WSEP) {
#pragma unroll
            for (int q = 0; q < 4; ++q) {
              float a = 0.0f;
#pragma unroll
              for (int k = 0; k < SX; ++k) a = __fmaf_rn(p.sv[k], xw[q + k], a);
              h[q] = a;
            }
          }
          static_for<SY>([&](auto KY) {
            constexpr int kyy = decltype(KY)::value;
            constexpr int slot_ = ((rs - kyy) % RS + RS) % RS;    // output row i - kyy
#pragma unroll
            for (int q = 0; q < 4; ++q) {
              float a = kyy == 0 ? 0.0f : acc[slot_][q];
              if constexpr (OP == K3_WSEP) {
                a = __fmaf_rn(p.su[kyy], h[q], a);
              } else if constexpr (OP == K3_WSTAR) {
                if constexpr (kyy == RY) {
#pragma unroll
                  for (int k = 0; k < SX; ++k) a = __fmaf_rn(p.wbox[kyy * SX + k], xw[q + k], a);
                } else {
                  a = __fmaf_rn(p.wbox[kyy * SX + RX], xw[q + RX], a);
                }
              } else {
#pragma unroll
                for (int k = 0; k < SX; ++k) a = __fmaf_rn(p.wbox[kyy * SX + k], xw[q + k], a);
              }
              acc[slot_][q] = a;
            }
            if constexpr (kyy == 2 * RY) store(i - 2 * RY, acc[slot_]);
          });
        } else {
#pragma unroll
          for (int q = 0; q < W; ++q) ra[rs][q] = xw[q];
          if constexpr (NIN > 1) {
            float4 c, e;
            fetch_row<XE>(row1, src1, yrow, it.x0, nx, lane, c, e);
            make_window<RX, XE>(c, e, lane, rb[rs], xs, pv);
            if (XE && yconst) {
#pragma unroll
              for (int q = 0; q < W; ++q) rb[rs][q] = pv;
            }
          }
          if (i >= 2 * RY) {
            // rows i-2RY .. i sit in slots (rs - 2RY + k) mod SY
            float wa[SY][W], wb[(NIN > 1) ? SY : 1][W];
#pragma unroll
            for (int k = 0; k < SY; ++k) {
              const int sl = ((rs - 2 * RY + k) % RS + RS) % RS;
#pragma unroll
              for (int q = 0; q < W; ++q) {
                wa[k][q] = ra[sl][q];
                if constexpr (NIN > 1) wb[k][q] = rb[sl][q];
              }
            }
            float v[4];
            static_for<4>([&](auto I) {
              constexpr int ii = decltype(I)::value;
              if constexpr (OP == K3_SRAD1) {
                v[ii] = op_srad1(RingAcc<RY, RX, ii>{wa}, p.prm);
              } else if constexpr (OP == K3_GRAD) {
                v[ii] = op_gradient(RingAcc<RY, RX, ii>{wa}, p.prm);
              } else if constexpr (OP == K3_HOT2D) {
                v[ii] = op_hotspot2d(RingAcc<RY, RX, ii>{wa}, RingAcc<RY, RX, ii>{wb}, p.prm);
              } else {
                v[ii] = op_srad2(RingAcc<RY, RX, ii>{wa}, RingAcc<RY, RX, ii>{wb}, p.prm);
              }
            });
            store(i - 2 * RY, v);
          }
        }
      };
      // U groups per iteration (RS rows): every row's slot is compile-time and
      // no shuffle sits under a data-dependent branch.  Rows past the item's
      // last input row (the tail of its last block) run too; their outputs
      // fall outside [0, nout) and are not stored.  After each group the warp
      // hands its slot back to the load cursor.
      for (int g0 = 0; g0 < it.ng; g0 += U) {
        static_for<U>([&](auto GI) {
          constexpr int gi = decltype(GI)::value;
          const int g = g0 + gi;
          mbar_wait(&bars[cs], (cphase >> cs) & 1u);
          cphase ^= 1u << cs;
          const float4* s0 = ring + cs * SLOT4;
          static_for<G>([&](auto J) {
            constexpr int j = decltype(J)::value;
            row(std::integral_constant<int, gi * G + j>{}, g * G + j, s0 + j * BX4, s0 + GROUP4 + j * BX4);
          });
          __syncwarp();
          if (++cs == S) cs = 0;
          --inflight;
          refill();
        });
      }
    };
    if (edge)
      sweep(std::true_type{});
    else
      sweep(std::false_type{});
    // next item: the one the load cursor already started, or a fresh ticket
    if (l_item != c_item) {
      c_item = l_item;
    } else {
      c_item = nitems;   // the load cursor found no further item
    }
    refill();
  }

  // last CTA out resets the launch slot's ticket counter (graph-replay safe)
  __syncthreads();
  if (threadIdx.x == 0) {
    __threadfence();
    const unsigned prev = atomicAdd(&g_launch[slot].c[1], 1u);
    if (prev == gridDim.x - 1) release_launch_slot(g_launch, slot);
  }
}

struct Launcher {
  const void* fn;
  int smem;
  int g;
  int wpc;
  int nin;
  int ctas_per_sm;
};

template <int OP, int RY, int RX, int G, int S, int NIN, int WPC, int MINB>
Launcher get_launcher() {
  static Launcher L{};
  static std::once_flag once;
  std::call_once(once, [] {
    using C = WCfg<G, S, NIN, WPC>;
    auto fn = k3_wsweep<OP, RY, RX, G, S, NIN, WPC, MINB>;
    cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, C::SMEM);
    int occ = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, fn, WPC * 32, C::SMEM) != cudaSuccess) occ = 1;
    cudaGetLastError();
    L = Launcher{reinterpret_cast<const void*>(fn), C::SMEM, G, WPC, NIN, occ > 0 ? occ : 1};
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

// (G rows per group, S groups in flight per warp, warps per CTA, min CTAs per SM)
#define K3_L1(OPV, RYV, RXV) get_launcher<OPV, RYV, RXV, 4, 6, 1, 8, 2>()
#define K3_L2(OPV, RYV, RXV) get_launcher<OPV, RYV, RXV, 4, 4, 2, 4, 3>()

// tuning hook (ATF role): LIFT_K3_VARIANT picks alternative
// (G, S, warps per CTA, min CTAs per SM) for the separable radius-2 Gaussian,
// SRAD1 and SRAD2; read per launch
template <int OPV, int RYV, int RXV, int NINV>
bool pick_variant(Launcher* L) {
  const char* e = getenv("LIFT_K3_VARIANT");
  const int v = e ? atoi(e) : 0;
  switch (v) {
    case 1: *L = get_launcher<OPV, RYV, RXV, 4, 4, NINV, 8, 3>(); return true;
    case 2: *L = get_launcher<OPV, RYV, RXV, 8, 3, NINV, 8, 2>(); return true;
    case 3: *L = get_launcher<OPV, RYV, RXV, 4, 8, NINV, 4, 3>(); return true;
    case 4: *L = get_launcher<OPV, RYV, RXV, 4, 3, NINV, 8, 4>(); return true;
    case 5: *L = get_launcher<OPV, RYV, RXV, 8, 4, NINV, 4, 3>(); return true;
    default: return false;
  }
}

bool pick(const StencilParams& p, Launcher* L) {
  const int ry = p.lo[1], rx = p.lo[2];
  if (p.op == OP_WEIGHTED && p.sep && ry == 2 && rx == 2 && pick_variant<K3_WSEP, 2, 2, 1>(L)) return true;
  if (p.op == OP_SRAD1 && pick_variant<K3_SRAD1, 1, 1, 1>(L)) return true;
  if (p.op == OP_SRAD2 && pick_variant<K3_SRAD2, 1, 1, 2>(L)) return true;
  if (p.op == OP_WEIGHTED) {
    const bool sep = p.sep != 0;
    const bool star = star2d(p, ry, rx);
#define K3_CASE(RYV, RXV)                                          \
  if (ry == RYV && rx == RXV) {                                    \
    if (sep) *L = K3_L1(K3_WSEP, RYV, RXV);                        \
    else if (star) *L = K3_L1(K3_WSTAR, RYV, RXV);                 \
    else *L = K3_L1(K3_WBOX, RYV, RXV);                            \
    return true;                                                   \
  }
    K3_CASE(1, 1)
    K3_CASE(2, 2)
    K3_CASE(1, 2)
    K3_CASE(2, 1)
#undef K3_CASE
    return false;
  }
  if (p.op == OP_SRAD1) { *L = K3_L1(K3_SRAD1, 1, 1); return true; }
  if (p.op == OP_GRADIENT) { *L = K3_L1(K3_GRAD, 1, 1); return true; }
  if (p.op == OP_SRAD2) { *L = K3_L2(K3_SRAD2, 1, 1); return true; }
  if (p.op == OP_HOTSPOT2D) { *L = K3_L2(K3_HOT2D, 1, 1); return true; }
  return false;
}

struct MapEntry {
  const float* base;
  int64_t nx, ny;
  int by;
  CUtensorMap map;
};

bool get_map(const float* base, int64_t nx, int64_t ny, int by, CUtensorMap* out, std::string* err) {
  thread_local MapEntry cache[16];
  thread_local int next = 0;
  for (auto& e : cache)
    if (e.base == base && e.nx == nx && e.ny == ny && e.by == by) {
      *out = e.map;
      return true;
    }
  MapEntry e{base, nx, ny, by, {}};
  if (!encode_tensor_map_3d(&e.map, base, nx, ny, 1, BX, (uint32_t)by, 1, err)) return false;
  cache[next] = e;
  next = (next + 1) % 16;
  *out = e.map;
  return true;
}

}  // namespace

bool wsweep2d_supported(const StencilParams& p, const float* in0, const float* in1, bool small) {
  // LIFT_K3=0 / =1 route every eligible plan to K1 / K3 (read per launch: A/B
  // tests and measurements).  Default: K3 for the non-separable weighted
  // stencils, Gradient and Hotspot2D on grids that fill the GPU (measured
  // faster than K1: J2D9 722 vs 676, Gradient 710 vs 648, Hotspot2D 492 vs
  // 445 Gpts/s at 8192^2); K1 keeps the separable Gaussian, SRAD1/SRAD2
  // (whose 128 x 48 / 128 x 32 tiles measured faster) and small grids.
  const char* e = getenv("LIFT_K3");
  const int mode = e ? (e[0] == '0' ? 0 : 1) : -1;
  if (mode == 0) return false;
  if (mode < 0) {
    if (small) return false;
    const bool pick = (p.op == OP_WEIGHTED && !p.sep) || p.op == OP_GRADIENT || p.op == OP_HOTSPOT2D;
    if (!pick) return false;
  }
  if (p.op == OP_SRAD) return false;                 // the fused SRAD iteration has its own kernel
  if (p.kind[2] == PAD_WRAP) return false;           // x wrap needs the far edge: K1's halo fix-up
  if (p.n[2] % 4 != 0) return false;                 // TMA row pitch
  if ((reinterpret_cast<uintptr_t>(in0) & 15u) || (in1 && (reinterpret_cast<uintptr_t>(in1) & 15u))) return false;
  return true;
}

cudaError_t launch_wsweep2d(const StencilParams& p, const float* in0, const float* in1, float* out,
                            cudaStream_t stream, int num_sms, std::string* err) {
  Launcher L;
  if (!pick(p, &L)) {
    *err = "wsweep2d: no instantiation";
    return cudaErrorNotSupported;
  }
  CUtensorMap m0{}, m1{};
  if (!get_map(in0, p.n[2], p.n[1], L.g, &m0, err)) return cudaErrorInvalidValue;
  if (L.nin > 1) {
    if (!get_map(in1, p.n[2], p.n[1], L.g, &m1, err)) return cudaErrorInvalidValue;
  } else {
    m1 = m0;
  }
  const float* s1 = L.nin > 1 ? in1 : in0;
  const int64_t nx = p.n[2], ny = p.n[1];
  const int nstrips = (int)((nx + TX - 1) / TX);
  const int64_t warps = (int64_t)num_sms * L.ctas_per_sm * L.wpc;
  // rows per item: ~8 items per warp for dynamic balance, at most 512, and
  // hc + 2R a multiple of the kernel's ring size so that every row is used
  // (LIFT_K3_HC forces a value: tests exercise multi-block sweeps on small grids)
  const int ry = p.lo[1];
  int64_t hc = (ny * nstrips + 8 * warps - 1) / (8 * warps);
  if (const char* e = getenv("LIFT_K3_HC")) hc = atoll(e);
  hc = std::min<int64_t>(std::max<int64_t>(hc, 1), 512);
  const int rsz = ((2 * ry + 1 + L.g - 1) / L.g) * L.g;     // the kernel's ring size RS
  hc = ((hc + 2 * ry + rsz - 1) / rsz) * rsz - 2 * ry;
  if (hc < 1) hc += rsz;
  const int64_t nchunks = (ny + hc - 1) / hc;
  const int64_t nitems = nchunks * nstrips;
  if (nitems > 0x7fffffff) return cudaErrorInvalidConfiguration;
  int64_t grid = (int64_t)num_sms * L.ctas_per_sm;
  const int64_t need = (nitems + L.wpc - 1) / L.wpc;
  if (grid > need) grid = need;
  int ns = nstrips, hci = (int)hc, ni = (int)nitems;
  void* args[] = {(void*)&p, (void*)&m0, (void*)&m1, (void*)&in0, (void*)&s1, (void*)&out, &ns, &hci, &ni};
  set_last_kernel("k3_wsweep");
  return launch_kernel(L.fn, dim3((unsigned)grid), dim3(L.wpc * 32), args, (size_t)L.smem, stream, true);
}

}  // namespace lift
