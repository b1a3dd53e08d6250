// kernel_sweep3d.cu — K2: the 3D stencil as a 2.5D sweep along z.
//
// slide_3 over a 3D grid.  Work items are (z-chunk, 128 x TY tile
// of the (y, x) plane) in chunk-major order; persistent CTAs (grid = SMs x
// resident CTAs) draw items from a dynamic ticket counter, so the CTAs in
// flight always work on neighbouring tiles of the same z range (their halo'd
// boxes overlap in L2) and there is no tail wave.
//
// Per CTA an elected producer thread streams the input planes of its items
// (z-R .. z_end+R-1 per item) through an S-stage shared-memory ring: one TMA
// tensor load per plane of a halo'd box of (128+8) x (TY+2R) floats (x from
// x0-4 so the centre columns stay 16-B aligned; y from y0-R), completing on
// the stage's mbarrier.  This is overlapped tiling with overlap
// size-step = 2R, staged in local (shared) memory.
//
// 8 consumer warps: lane l of warp w owns 4 consecutive x outputs of TY/8
// rows.  The centre float4 of every plane is read from shared memory once,
// when the plane lands, into a per-thread register ring of 2R+1 planes (the
// z-neighbours); when plane z is the centre, its y-neighbours are 128-bit
// shared loads and its in-row neighbours come from the adjacent lanes by warp
// shuffles (lanes 0/31 read the halo columns).  A plane's stage is released as
// soon as it has served as the centre, so the ring needs only R+1 live stages
// plus prefetch.  Results leave as one st.global.v4 per lane and row.
//
// pad is folded into index computation: the producer remaps the
// plane index (or marks a constant plane, which is never loaded); inside a
// plane, clamp / mirror / reflect / constant rows are redirected to the
// remapped box row, and out-of-grid x taps are selected from the lane's own
// registers; only WRAP in x or y rewrites the halo cells in shared memory from
// global memory (halo.cuh).  f goes through ops.cuh: every output has exactly
// the bits K0 computes.
#include <cuda.h>
#include <cuda_runtime.h>

#include <algorithm>
#include <atomic>
#include <climits>
#include <cstdlib>
#include <mutex>
#include <string>
#include <type_traits>

#include "common.cuh"
#include "halo.cuh"
#include "launch.hpp"
#include "ops.cuh"
#include "slots.cuh"
#include "tma.cuh"

namespace lift {
namespace {

constexpr int TX = 128;        // outputs per tile row: 32 lanes x float4
constexpr int XH = 4;          // halo columns loaded on each side (>= R, keeps 16-B alignment)
constexpr int BX = TX + 2 * XH;
constexpr int NW = 8;          // consumer warps
constexpr int NCONS = NW * 32;
constexpr unsigned FULL = 0xffffffffu;
// dynamic work counters, one slot per running launch (slots.cuh): c[0] item
// ticket, c[1] CTAs done, c[2..3] finished boundary-chunk items (fused step)
__device__ LaunchSlot g_launch[kLaunchSlots];

// fused step: boundary chunks first (item order: chunk 0, chunk last, then the rest)
__device__ __forceinline__ int chunk_of(int c, int nchunk, bool fused) {
  if (!fused || nchunk <= 2) return c;
  return c == 0 ? 0 : (c == 1 ? nchunk - 1 : c - 1);
}

// first plane (relative to reg0) of z-chunk c: the first n1 chunks hold zc
// planes, the rest zc2 (guided schedule: the last waves of items are short,
// so the launch's tail — CTAs still finishing their last item while the
// others idle — is short too)
__device__ __forceinline__ int64_t chunk_z0(int c, int zc, int n1, int zc2) {
  return c < n1 ? (int64_t)c * zc : (int64_t)n1 * zc + (int64_t)(c - n1) * zc2;
}

enum K2Op { K2_WSTAR = 0, K2_HOTSPOT = 1, K2_ACOUSTIC = 2, K2_WBOX = 3, K2_WBOX19 = 4 };
// 3x3x3 box weights; K2_WBOX19: the 8 corner taps are zero (Poisson 19-point)
// and are skipped at compile time (19 instead of 27 FMAs per point)
constexpr bool is_box(int op) { return op == K2_WBOX || op == K2_WBOX19; }

template <int R, int RPW, int S, int PSN>
struct Cfg {
  static constexpr int TY = NW * RPW;
  static constexpr int BY = TY + 2 * R;
  static constexpr int TX_BYTES = BX * BY * 4;
  static constexpr int STAGE_FLOATS = ((TX_BYTES + 127) / 128) * 128 / 4;
  static constexpr int PS = PSN;                        // point-wise ring slots (0: no point-wise grid)
  static constexpr int PW_BYTES = TX * TY * 4;
  static constexpr int PW_FLOATS = TX * TY;
  static constexpr int SMEM = S * STAGE_FLOATS * 4 + PS * PW_BYTES + 2 * (S + PS + 4) * 8 + (2 * S + 4) * 4 + 256;
};

template <int R>
struct Win {
  float x[4 + 2 * R];   // centre row, x offsets -R .. 3+R
  float ym[R][4];
  float yp[R][4];
  float zm[R][4];
  float zp[R][4];
};

template <int R, int I>
struct WinAcc {
  const Win<R>& w;
  template <int DZ, int DY, int DX>
  __device__ __forceinline__ float at() const {
    static_assert((DZ != 0) + (DY != 0) + (DX != 0) <= 1, "star access only");
    if constexpr (DZ < 0) return w.zm[-DZ - 1][I];
    else if constexpr (DZ > 0) return w.zp[DZ - 1][I];
    else if constexpr (DY < 0) return w.ym[-DY - 1][I];
    else if constexpr (DY > 0) return w.yp[DY - 1][I];
    else return w.x[I + R + DX];
  }
};

__device__ __forceinline__ void set4(float (&d)[4], float4 v) {
  d[0] = v.x; d[1] = v.y; d[2] = v.z; d[3] = v.w;
}

template <int OP, int R, int I>
__device__ __forceinline__ float eval(const StencilParams& p, const Win<R>& w, const float4& pw, int gz, int gy,
                                      int gx0) {
  WinAcc<R, I> a{w};
  if constexpr (OP == K2_WSTAR) {
    return op_weighted<R, R, R, true>(a, p.wbox);
  } else if constexpr (OP == K2_HOTSPOT) {
    return op_hotspot3d(a, f4get(pw, I), p.prm);
  } else {
    const int K = acoustic_K<R, int>(gz, gy, gx0 + I, (int)p.gnz, (int)p.n[1], (int)p.n[2]);
    return op_acoustic<R>(a, f4get(pw, I), K, p.prm);
  }
}

// Out-of-grid x taps of a lane's window (x = xo - R + m outside [0, nx)) for
// CLAMP / MIRROR / REFLECT / CONSTANT: the remapped tap lies in the lane's own
// float4 (R <= 2 < 4 <= nx), selected without dynamic register indexing.
__device__ __forceinline__ float pick4(int s, const float4& c, float pv) {
  return s < 0 ? pv : (s == 0 ? c.x : (s == 1 ? c.y : (s == 2 ? c.z : c.w)));
}

template <int OP, int R, int RPW, int S, bool ZC, bool FZ, int PSN>
__global__ void __launch_bounds__(NCONS + 32, (!is_box(OP) && (R == 1 || RPW == 1)) ? 3 : 2)
    k2_sweep(const __grid_constant__ StencilParams p, const __grid_constant__ CUtensorMap tmap,
             const __grid_constant__ CUtensorMap pwmap, const float* __restrict__ src, float* out, int ntx,
             int nty, int zc, int nchunk, int n1, int zc2) {
  using C = Cfg<R, RPW, S, (OP == K2_HOTSPOT || OP == K2_ACOUSTIC) ? PSN : 0>;
  constexpr bool PW = OP == K2_HOTSPOT || OP == K2_ACOUSTIC;           // a point-wise zipped grid (Hotspot P, Acoustic prev)
  constexpr int PS = C::PS;                     // point-wise ring slots
  constexpr int QN = 4;                         // item queue between the two producer lanes
  constexpr int PWF4 = C::PW_FLOATS / 4;
  constexpr int TY = C::TY;
  constexpr int SF4 = C::STAGE_FLOATS / 4;      // stage size in float4
  constexpr int BX4 = BX / 4;
  // dynamic smem (no static smem in this kernel, so it starts the CTA's window):
  // [S plane stages][PS point-wise slots][full S][empty S][pwfull PS][pwempty PS][stage_item S][stage_const S]
  extern __shared__ __align__(128) float4 dsm4[];
  uint64_t* full = reinterpret_cast<uint64_t*>(dsm4 + S * SF4 + PS * PWF4);
  uint64_t* empty = full + S;
  uint64_t* pwfull = empty + S;
  uint64_t* pwempty = pwfull + PS;
  uint64_t* itemfull = pwempty + PS;
  uint64_t* itemempty = itemfull + QN;
  int* stage_item = reinterpret_cast<int*>(itemempty + QN);
  int* stage_const = stage_item + S;
  int* item_q = stage_const + S;
  int* slot_sm = item_q + QN;

  const int ntile = ntx * nty;
  const int nitems = ntile * nchunk;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;

  if (threadIdx.x == 0) {
    for (int s = 0; s < S; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NW);
    }
    for (int s = 0; s < PS; ++s) {
      mbar_init(&pwfull[s], 1);
      mbar_init(&pwempty[s], NW);
    }
    for (int s = 0; s < QN; ++s) {
      mbar_init(&itemfull[s], 1);
      mbar_init(&itemempty[s], 1);
    }
    fence_mbar_init();
    *slot_sm = claim_launch_slot(g_launch);
  }
  __syncthreads();
  const int slot = *slot_sm;
  pdl_launch_dependents();   // PDL: let the next launch ramp up now
  pdl_wait();                // ... and wait for the previous one before any global access

  if (warp == NW) {
    // ---------------- producers ----------------
    // lane 0: items from the ticket counter, one TMA box per input plane;
    // lane 1 (point-wise ops): the point-wise box of every output plane, fed
    // the item sequence through a small queue so that a full point-wise ring
    // never holds back the plane prefetch
    if (lane == 0) {
      prefetch_tmap(&tmap);
      int s = 0;
      uint32_t pass = 0;
      int q = 0;
      uint32_t qpass = 0;
      while (true) {
        const int item = (int)atomicAdd(&g_launch[slot].c[0], 1u);
        const bool done = item >= nitems;
        if constexpr (PW) {
          if (qpass > 0) mbar_wait(&itemempty[q], (qpass - 1) & 1);
          item_q[q] = done ? -1 : item;
          mbar_arrive(&itemfull[q]);
          if (++q == QN) { q = 0; ++qpass; }
        }
        int nload = 1, x0 = 0, y0 = 0;
        int64_t zs = 0;
        if (!done) {
          const int chunk = chunk_of(item / ntile, nchunk, FZ && p.fused_step), tile = item % ntile;
          x0 = (tile % ntx) * TX;
          y0 = (tile / ntx) * TY;
          zs = p.reg0 + chunk_z0(chunk, zc, n1, zc2);
          const int64_t ze = min(zs + (int64_t)(chunk < n1 ? zc : zc2), p.reg1);
          nload = (int)(ze - zs) + 2 * R;
          // fused step: the ghost planes of this chunk must hold the neighbours'
          // previous step before the TMA reads them
          if constexpr (FZ) {
            bool waited = false;
            if (chunk == 0 && p.wait_lo) {
              spin_until_bounded(p.wait_lo, p.wait_value, p.wait_timeout_ns, p.fault, kFaultWaitLo);
              waited = true;
            }
            if (chunk == nchunk - 1 && p.wait_hi) {
              spin_until_bounded(p.wait_hi, p.wait_value, p.wait_timeout_ns, p.fault, kFaultWaitHi);
              waited = true;
            }
            if (waited) asm volatile("fence.proxy.async.global;" ::: "memory");
          }
        }
        // a "done" marker occupies one stage so the consumers see it in order
        for (int i = 0; i < nload; ++i) {
          if (pass > 0) mbar_wait(&empty[s], (pass - 1) & 1);
          const int64_t lz = done ? -1 : plane_of(p, p.z_off + zs - R + i);
          if (i == 0) stage_item[s] = done ? -1 : item;
          stage_const[s] = lz < 0;
          if (!done && (lz >= 0 || !ZC)) {
            // a zero value-pad plane (kind CONSTANT, pad_value 0, !ZC) is loaded at
            // z = -1: entirely out of bounds, so TMA fills it with zeros (no HBM bytes)
            mbar_arrive_expect_tx(&full[s], C::TX_BYTES);
            tma_load_3d(dsm4 + s * SF4, &tmap, &full[s], x0 - XH, y0 - R, lz >= 0 ? (int)lz : -1);
          } else {
            mbar_arrive(&full[s]);   // non-zero constant plane (ZC) or end marker: nothing to load
          }
          if (++s == S) { s = 0; ++pass; }
        }
        if (done) break;
      }
    } else if (PW && lane == 1) {
      prefetch_tmap(&pwmap);
      int ps = 0, q = 0;
      uint32_t ppass = 0, qpass = 0;
      while (true) {
        mbar_wait(&itemfull[q], qpass & 1);
        const int item = item_q[q];
        mbar_arrive(&itemempty[q]);
        if (++q == QN) { q = 0; ++qpass; }
        if (item < 0) break;
        const int chunk = chunk_of(item / ntile, nchunk, FZ && p.fused_step), tile = item % ntile;
        const int x0 = (tile % ntx) * TX, y0 = (tile / ntx) * TY;
        const int64_t zs = p.reg0 + chunk_z0(chunk, zc, n1, zc2);
        const int nzc = (int)(min(zs + (int64_t)(chunk < n1 ? zc : zc2), p.reg1) - zs);
        for (int j = 0; j < nzc; ++j) {
          if (ppass > 0) mbar_wait(&pwempty[ps], (ppass - 1) & 1);
          mbar_arrive_expect_tx(&pwfull[ps], C::PW_BYTES);
          tma_load_3d(dsm4 + S * SF4 + ps * PWF4, &pwmap, &pwfull[ps], x0, y0, (int)(zs + j + p.ghost));
          if (++ps == PS) { ps = 0; ++ppass; }
        }
      }
    }
  } else {
    // ---------------- consumers ----------------
    const int nx = (int)p.n[2], ny = (int)p.n[1];
    const int kx = p.kind[2], ky = p.kind[1];
    const float pv = p.pad_value;
    const float4 pv4 = make_float4(pv, pv, pv, pv);
    // WRAP and non-zero CONSTANT in x/y rewrite the halo cells in shared memory;
    // zero CONSTANT is TMA's out-of-bounds fill; CLAMP/MIRROR/REFLECT are folded
    // into row offsets (y) and register selects (x)
    const bool wrap_fix = (kx == PAD_WRAP || ky == PAD_WRAP) ||
                          ((kx == PAD_CONSTANT || ky == PAD_CONSTANT) && pv != 0.0f);
    // float4 offset (within a stage) of this thread's first row, centre column
    const int roff4 = (warp * RPW + R) * BX4 + XH / 4 + lane;
    // CLAMP / MIRROR / REFLECT in x: out-of-grid x taps are read from the
    // remapped in-grid column of the same row (address folded in per item)
    const bool x_remap = !wrap_fix && kx != PAD_CONSTANT;
    const float* dsf = reinterpret_cast<const float*>(dsm4);
    // Acoustic interior constants: x part of K when all 4 x-neighbour sets are
    // in the domain, and the centre coefficient 2 - l2*K at K = 6R
    constexpr int kx_full = (2 * R) * 0x1111;
    const float a_int = __fsub_rn(2.0f, __fmul_rn(p.prm[0], (float)(6 * R)));
    int sn = 0;            // stage of the next load to wait for
    uint32_t pn = 0;       // its pass (barrier phase parity)
    int psc = 0;           // point-wise ring slot of the current output plane
    uint32_t ppc = 0;
    while (true) {
      mbar_wait(&full[sn], pn & 1);
      const int item = stage_item[sn];
      if (item < 0) {
        __syncwarp();
        if (lane == 0) mbar_arrive(&empty[sn]);
        break;
      }
      const int chunk = chunk_of(item / ntile, nchunk, FZ && p.fused_step), tile = item % ntile;
      const int x0 = (tile % ntx) * TX;
      const int y0 = (tile / ntx) * TY;
      const int64_t zs = p.reg0 + chunk_z0(chunk, zc, n1, zc2);
      const int nzc = (int)(min(zs + (int64_t)(chunk < n1 ? zc : zc2), p.reg1) - zs);
      const int xo = x0 + 4 * lane;
      const bool x_ok = xo < nx;
      const bool y_edge = (y0 < R) || (y0 + TY + R > ny);
      const bool x_edge = (x0 == 0) || (x0 + TX + R > nx);
      const bool fix = wrap_fix && (x_edge || y_edge);
      const bool yr = !wrap_fix && ky != PAD_CONSTANT && y_edge;
      // Edge items (the tile or its halo touches the grid boundary) run the
      // general loop body; interior items a specialised copy with compile-time
      // row offsets, no pad logic and no store predicates.
      // x halo taps: lanes 1..31 take x-1..x-R from the lane below by shuffle,
      // x+1..x+R from the lane above.  Interior: lane 0 / lane 31 take them from
      // the halo float4 of the row.  Edge: lane 0 reads them from shared memory
      // at lrel (floats, relative to its centre element), lane 31 and the lane
      // holding the last in-grid column at rrel — for CLAMP / MIRROR / REFLECT
      // the remapped in-grid column of the same row; lanes that do not use the
      // read get lane 0's / lane 31's address (a broadcast).
      const bool x_last = x_remap && xo + 4 == nx;
      const bool use_r = lane == 31 || x_last;
      int lrel[R], rrel[R];
#pragma unroll
      for (int k = 1; k <= R; ++k) {
        lrel[k - 1] = (x_remap && x0 == 0 && lane == 0) ? (int)pad_remap(-k, nx, kx) : -k - 4 * lane;
        rrel[k - 1] = x_last ? (int)pad_remap(nx - 1 + k, nx, kx) - xo : TX - 1 + k - 4 * lane;
      }
      // float4 offset of the halo float4 of a row relative to the lane's centre float4
      const int eo4 = (lane == 0 ? 0 : (XH + TX) / 4) - XH / 4 - lane;
      // Acoustic: x part of the in-domain neighbour count of the lane's 4
      // outputs, packed 4 bits each (computed once per item)
      int kxp = 0;
      // and its y part per output row (the z part comes per plane): K = Kz +
      // Ky + Kx with one add per row instead of 4R compares
      int kyr[RPW];
      if constexpr (OP == K2_ACOUSTIC) {
#pragma unroll
        for (int i = 0; i < 4; ++i) {
          int kxi = 0;
#pragma unroll
          for (int o = 1; o <= R; ++o) kxi += (xo + i - o >= 0) + (xo + i + o < nx);
          kxp |= kxi << (4 * i);
        }
#pragma unroll
        for (int jj = 0; jj < RPW; ++jj) {
          const int gy = y0 + warp * RPW + jj;
          int k = 0;
#pragma unroll
          for (int o = 1; o <= R; ++o) k += (gy - o >= 0) + (gy + o < ny);
          kyr[jj] = k;
        }
      }
      // float4 offset of the warp's row d - R (d = 0 .. RPW-1+2R) relative to
      // its first row, with the y pad redirect folded in (edge items)
      int rowo[RPW + 2 * R];
#pragma unroll
      for (int d = 0; d < RPW + 2 * R; ++d) {
        const int gy = y0 + warp * RPW + d - R;
        rowo[d] = (d - R) * BX4;
        if (yr && (gy < 0 || gy >= ny))
          rowo[d] = (min(max((int)pad_remap(gy, ny, ky) - y0 + R, 0), C::BY - 1) - (warp * RPW + R)) * BX4;
      }
      // Stages of the 2R+1 planes around the current output plane z: zst[k]
      // holds plane z - R + k as the float4 offset of its stage (sn * SF4), or
      // -1 - sn * SF4 for a non-zero constant value plane (ZC; zero planes are
      // TMA out-of-bounds fills and read like any other stage)
      int zst[2 * R + 1];
      auto zenc = [&](int st) { return (ZC && stage_const[st]) ? -1 - st * SF4 : st * SF4; };
      auto zdec = [&](int v) { return (v < 0 ? -1 - v : v) / SF4; };
      // WRAP / non-zero constant: rewrite a plane's out-of-grid halo cells as
      // soon as it arrives (no warp has read that stage since its TMA landed),
      // so every plane of a window — not only the centre — is complete
      // (box windows read the halo of every plane: fix each plane on arrival;
      // star windows read only the centre plane's halo: fix the centre)
      constexpr bool FIX_ON_ARRIVAL = is_box(OP);
      auto fix_plane = [&](int stage, int64_t gzp) {
        if (stage_const[stage]) return;
        fixup_tile<R, R, XH, BX, C::BY, NCONS>(p, reinterpret_cast<float*>(dsm4 + stage * SF4), src,
                                               plane_of(p, gzp), x0, y0, threadIdx.x);
        fence_proxy_async_smem();
      };
      float* orow = out + ((zs + p.ghost) * p.plane + (int64_t)(y0 + warp * RPW) * nx + xo);

      auto plane_loop = [&](auto edge_tag) {
        constexpr bool EDGE = decltype(edge_tag)::value;
        auto RO = [&](int d) { return EDGE ? rowo[d] : (d - R) * BX4; };
        // the x-window (offsets -R .. 3+R) of the row whose centre float4 is at
        // a (c = its value; cz: a constant value plane)
        auto xwin = [&](int a, const float4& c, bool cz, float (&xw)[4 + 2 * R]) {
          const float cv[4] = {c.x, c.y, c.z, c.w};
          float4 e = pv4;
          if (!EDGE && !(ZC && cz)) e = dsm4[a + eo4];
          const float ev[4] = {e.x, e.y, e.z, e.w};
#pragma unroll
          for (int k = 1; k <= R; ++k) {
            float l = __shfl_up_sync(FULL, cv[4 - k], 1);
            float r = __shfl_down_sync(FULL, cv[k - 1], 1);
            if constexpr (EDGE) {
              const float hl = (ZC && cz) ? pv : dsf[a * 4 + lrel[k - 1]];
              const float hr = (ZC && cz) ? pv : dsf[a * 4 + rrel[k - 1]];
              if (lane == 0) l = hl;
              if (use_r) r = hr;
            } else {
              if (lane == 0) l = ev[4 - k];
              if (lane == 31) r = ev[k - 1];
            }
            xw[R - k] = l;
            xw[R + 3 + k] = r;
          }
#pragma unroll
          for (int i = 0; i < 4; ++i) xw[R + i] = cv[i];
        };
        // 3x3x3 box: running accumulators along z.  Each arriving plane q is read
        // once (rows -1 .. RPW, one x-window each) and its taps go to three
        // outputs: q-1 (kz = 2, completes it), q (kz = 1) and q+1 (kz = 0, starts
        // it).  Every output's FMA chain still runs over its 27 taps in
        // row-major (kz, ky, kx) order from 0 — K0's order, so the bits agree.
        float P1[RPW][4], P0[RPW][4];     // partial sums of outputs q and q+1
        if constexpr (is_box(OP)) {
#pragma unroll
          for (int jj = 0; jj < RPW; ++jj)
#pragma unroll
            for (int i = 0; i < 4; ++i) P1[jj][i] = P0[jj][i] = 0.0f;
        }
        auto box_plane = [&](int az, float (&O)[RPW][4]) {
          const bool cz = ZC && az < 0;
          const int sb = cz ? 0 : az;
          float N1[RPW][4], N0[RPW][4];
#pragma unroll
          for (int jj = 0; jj < RPW; ++jj)
#pragma unroll
            for (int i = 0; i < 4; ++i) {
              O[jj][i] = P1[jj][i];
              N1[jj][i] = P0[jj][i];
              N0[jj][i] = 0.0f;
            }
#pragma unroll
          for (int d = 0; d < RPW + 2; ++d) {
            const int a = sb + roff4 + RO(d);
            const float4 c2 = cz ? pv4 : dsm4[a];
            float w6[4 + 2 * R];
            xwin(a, c2, cz, w6);
#pragma unroll
            for (int jj = 0; jj < RPW; ++jj) {
              const int kyy = d - jj;
              if (kyy < 0 || kyy > 2) continue;
#pragma unroll
              for (int kxx = 0; kxx < 3; ++kxx) {
                const float w2 = p.wbox[(2 * 3 + kyy) * 3 + kxx];
                const float w1 = p.wbox[(1 * 3 + kyy) * 3 + kxx];
                const float w0 = p.wbox[(0 * 3 + kyy) * 3 + kxx];
                // corner taps (kz, ky, kx all off-centre) of the 19-point pattern
                const bool corner = OP == K2_WBOX19 && kyy != 1 && kxx != 1;
#pragma unroll
                for (int i = 0; i < 4; ++i) {
                  if (!corner) O[jj][i] = __fmaf_rn(w2, w6[i + kxx], O[jj][i]);
                  N1[jj][i] = __fmaf_rn(w1, w6[i + kxx], N1[jj][i]);
                  if (!corner) N0[jj][i] = __fmaf_rn(w0, w6[i + kxx], N0[jj][i]);
                }
              }
            }
          }
#pragma unroll
          for (int jj = 0; jj < RPW; ++jj)
#pragma unroll
            for (int i = 0; i < 4; ++i) {
              P1[jj][i] = N1[jj][i];
              P0[jj][i] = N0[jj][i];
            }
        };
        // the first 2R planes of the chunk
#pragma unroll
        for (int k = 0; k < 2 * R; ++k) {
          if (k > 0) mbar_wait(&full[sn], pn & 1);
          zst[k] = zenc(sn);
          if constexpr (FIX_ON_ARRIVAL && EDGE) {
            if (fix) {
              fix_plane(sn, p.z_off + zs - R + k);
              named_bar_sync(1, NCONS);
            }
          }
          if (++sn == S) { sn = 0; ++pn; }
          if constexpr (is_box(OP)) {
            float O[RPW][4];
            box_plane(zst[k], O);          // O: not an output yet
          }
        }
        for (int j = 0; j < nzc; ++j) {
          mbar_wait(&full[sn], pn & 1);
          zst[2 * R] = zenc(sn);
          const int64_t z = zs + j;                  // local output plane
          const int gz = (int)(p.z_off + z);
          int kzp = 0;             // Acoustic: z part of K for this output plane
          if constexpr (OP == K2_ACOUSTIC) {
#pragma unroll
            for (int o = 1; o <= R; ++o) kzp += (gz - o >= 0) + (gz + o < (int)p.gnz);
          }
          if constexpr (FIX_ON_ARRIVAL && EDGE) {
            if (fix) {
              fix_plane(sn, p.z_off + z + R);
              named_bar_sync(1, NCONS);
            }
          }
          if (++sn == S) { sn = 0; ++pn; }
          const int cbase = zst[R];                   // the centre plane is inside the grid
          if constexpr (!FIX_ON_ARRIVAL && EDGE) {
            if (fix) {
              // all warps are past the previous plane (which read this stage as its
              // z+1 neighbour, including the padding lanes/rows of ragged tiles)
              named_bar_sync(1, NCONS);
              fixup_tile<R, R, XH, BX, C::BY, NCONS>(p, reinterpret_cast<float*>(dsm4 + cbase), src,
                                                     plane_of(p, (int64_t)gz), x0, y0, threadIdx.x);
              fence_proxy_async_smem();
              named_bar_sync(1, NCONS);
            }
          }
          // point-wise input of this output plane: its own TMA ring (no halo)
          if constexpr (PW) mbar_wait(&pwfull[psc], ppc & 1);
          // box: plane z+1 completes output z
          float BO[RPW][4];
          if constexpr (is_box(OP)) box_plane(zst[2], BO);
          // star ops: rows -R .. RPW-1+R of the centre plane, each read once
          float4 cr[RPW + 2 * R];
          if constexpr (!is_box(OP)) {
#pragma unroll
            for (int d = 0; d < RPW + 2 * R; ++d) cr[d] = dsm4[cbase + roff4 + RO(d)];
          }
#pragma unroll
          for (int jj = 0; jj < RPW; ++jj) {
            const int rr = warp * RPW + jj;
            const int gy = y0 + rr;
            const bool ok = EDGE ? (x_ok && gy < ny) : true;
            float4 pw = make_float4(0.f, 0.f, 0.f, 0.f);
            if constexpr (PW) pw = dsm4[S * SF4 + psc * PWF4 + (warp * RPW + jj) * (TX / 4) + lane];
            const int rb = roff4 + jj * BX4;          // natural row offset within a stage
            auto zrow = [&](int k) -> float4 {       // centre float4 of plane z + k
              const int a = zst[R + k];
              if constexpr (ZC) return a < 0 ? pv4 : dsm4[a + rb];
              return dsm4[a + rb];
            };
            float4 res;
            if constexpr (is_box(OP)) {
              res = make_float4(BO[jj][0], BO[jj][1], BO[jj][2], BO[jj][3]);
            } else {
              float xw[4 + 2 * R];                    // centre row, x offsets -R .. 3+R
              xwin(cbase + roff4 + RO(jj + R), cr[jj + R], false, xw);
              if constexpr (OP == K2_ACOUSTIC) {
                // ordered neighbour sum (acoustic_sum's row-major order), accumulated
                // as the taps are loaded: z-R..z-1, y-R..y-1, x-R..x-1, x+1..x+R,
                // y+1..y+R, z+1..z+R
                float sm[4];
                bool first = true;
                auto add4 = [&](const float4& v) {
                  const float vv[4] = {v.x, v.y, v.z, v.w};
#pragma unroll
                  for (int i = 0; i < 4; ++i) sm[i] = first ? vv[i] : __fadd_rn(sm[i], vv[i]);
                  first = false;
                };
#pragma unroll
                for (int k = R; k >= 1; --k) add4(zrow(-k));
#pragma unroll
                for (int k = R; k >= 1; --k) add4(cr[jj + R - k]);
#pragma unroll
                for (int k = R; k >= 1; --k) add4(make_float4(xw[0 + R - k], xw[1 + R - k], xw[2 + R - k], xw[3 + R - k]));
#pragma unroll
                for (int k = 1; k <= R; ++k) add4(make_float4(xw[0 + R + k], xw[1 + R + k], xw[2 + R + k], xw[3 + R + k]));
#pragma unroll
                for (int k = 1; k <= R; ++k) add4(cr[jj + R + k]);
#pragma unroll
                for (int k = 1; k <= R; ++k) add4(zrow(k));
                const int Kzy = kzp + kyr[jj];
                const float pwv[4] = {pw.x, pw.y, pw.z, pw.w};
                float rv[4];
                if (Kzy == 4 * R && kxp == kx_full) {
                  // all 4 points interior (K = 6R): cf1 = cf2 = 1 and 2 - l2*K is a
                  // per-launch constant; the operations left are acoustic_combine's
                  // (the product by cf1 = 1 is exact), so the bits are unchanged
#pragma unroll
                  for (int i = 0; i < 4; ++i) {
                    float t = __fmul_rn(a_int, xw[R + i]);
                    t = __fmaf_rn(p.prm[0], sm[i], t);
                    rv[i] = __fmaf_rn(-1.0f, pwv[i], t);
                  }
                } else {
#pragma unroll
                  for (int i = 0; i < 4; ++i)
                    rv[i] = acoustic_combine<R>(sm[i], xw[R + i], pwv[i], Kzy + ((kxp >> (4 * i)) & 15), p.prm);
                }
                res = make_float4(rv[0], rv[1], rv[2], rv[3]);
              } else {
                Win<R> w;
#pragma unroll
                for (int i = 0; i < 4 + 2 * R; ++i) w.x[i] = xw[i];
#pragma unroll
                for (int k = 1; k <= R; ++k) {
                  set4(w.ym[k - 1], cr[jj + R - k]);
                  set4(w.yp[k - 1], cr[jj + R + k]);
                  set4(w.zm[k - 1], zrow(-k));
                  set4(w.zp[k - 1], zrow(k));
                }
                res.x = eval<OP, R, 0>(p, w, pw, gz, gy, xo);
                res.y = eval<OP, R, 1>(p, w, pw, gz, gy, xo);
                res.z = eval<OP, R, 2>(p, w, pw, gz, gy, xo);
                res.w = eval<OP, R, 3>(p, w, pw, gz, gy, xo);
              }
            }
            if (ok) {
              stg128(orow + jj * nx, res);
              if constexpr (FZ && EDGE) {
                // fused halo put: boundary planes also go to the neighbour's ghosts
                // (items of the boundary chunks run this general loop body)
                if (z < p.ghost && p.put_lo) stg128(p.put_lo + z * p.plane + (int64_t)gy * nx + xo, res);
                if (z >= p.n[0] - p.ghost && p.put_hi)
                  stg128(p.put_hi + (z - (p.n[0] - p.ghost)) * p.plane + (int64_t)gy * nx + xo, res);
              }
            }
          }
          orow += p.plane;
          // plane z - R is no longer needed (pre-chunk planes included)
          __syncwarp();
          if (lane == 0) {
            mbar_arrive(&empty[zdec(zst[0])]);
            if constexpr (PW) mbar_arrive(&pwempty[psc]);
          }
          if constexpr (PW) {
            if (++psc == PS) { psc = 0; ++ppc; }
          }
#pragma unroll
          for (int k = 0; k < 2 * R; ++k) zst[k] = zst[k + 1];
        }
      };
      // fused halo put: only the items of the first / last chunk store into the
      // neighbours' ghosts; they take the general (EDGE) body, every other
      // item the interior one without the put checks
      const bool put_item = FZ && (p.put_lo || p.put_hi) && (zs < p.ghost || zs + nzc > p.n[0] - p.ghost);
      if (x_edge || y_edge || put_item) plane_loop(std::true_type{});
      else plane_loop(std::false_type{});
      // the chunk's last 2R planes (z_end - R .. z_end + R - 1) are still held
      __syncwarp();
      if (lane == 0) {
#pragma unroll
        for (int k = 0; k < 2 * R; ++k) mbar_arrive(&empty[zdec(zst[k])]);
        // fused step: when every warp of every tile of a boundary chunk is done,
        // publish its peer stores and raise that neighbour's flag
        if (FZ && p.fused_step) {
          const unsigned need = (unsigned)ntile * NW;
          if (chunk == 0 && p.sig_lo) {
            __threadfence_system();
            if (atomicAdd(&g_launch[slot].c[2], 1u) == need - 1) {
              __threadfence_system();
              st_release_sys(p.sig_lo, p.sig_value);
            }
          }
          if (chunk == nchunk - 1 && p.sig_hi) {
            __threadfence_system();
            if (atomicAdd(&g_launch[slot].c[3], 1u) == need - 1) {
              __threadfence_system();
              st_release_sys(p.sig_hi, p.sig_value);
            }
          }
        }
      }
    }
  }
  // last CTA out resets the launch slot's counters (graph-replay safe) and,
  // for a fused halo put, publishes the ghost planes to the neighbours
  const bool puts = FZ && (p.put_lo || p.put_hi);
  if (puts) __threadfence_system();     // this thread's peer stores before the CTA's arrival
  __syncthreads();
  if (threadIdx.x == 0) {
    __threadfence();
    const unsigned prev = atomicAdd(&g_launch[slot].c[1], 1u);
    if (prev == gridDim.x - 1) {
      if (puts && !p.fused_step) {
        __threadfence_system();
        if (p.sig_lo) st_release_sys(p.sig_lo, p.sig_value);
        if (p.sig_hi) st_release_sys(p.sig_hi, p.sig_value);
      }
      release_launch_slot(g_launch, slot);
    }
  }
}

// ---------------------------------------------------------------------------
// K2T: two time steps per pass (temporal blocking) for the
// weighted 7-point star with CLAMP / MIRROR / REFLECT boundaries.
//
// X_t planes stream through the same TMA ring as K2 (box (128+8) x (16+2) at
// (x0-8, y0-2)); for each plane yz the 8 warps compute X_{t+1} on the
// extended 128 x 16 tile (columns x0-4 .. x0+123, rows y0-1 .. y0+14) into a
// 4-slot shared-memory ring, then — one barrier later — X_{t+2} on the inner
// 120 x 14 tile of plane yz-1 from the three ring planes.  Every value goes
// through op_weighted, so the result is bitwise equal to two single steps.
// pad applies to X_{t+1} as to any grid: its out-of-grid rows/columns are
// redirected to the remapped in-grid ones, and a plane outside the grid
// (global z = -1 or nz) aliases the remapped plane's ring slot.
// ---------------------------------------------------------------------------
constexpr int T2_TXO = 120;     // output columns per tile (lanes 1..30)
constexpr int T2_TYO = 14;      // output rows per tile (Y rows 1..14)
constexpr int T2_TY = 16;       // X_{t+1} rows per tile (2 per warp)
constexpr int T2_BY = T2_TY + 2;
constexpr int T2_YF4 = T2_TY * (TX / 4);   // float4 per X_{t+1} plane slot

template <int S>
struct CfgT2 {
  static constexpr int TX_BYTES = BX * T2_BY * 4;
  static constexpr int STAGE_FLOATS = ((TX_BYTES + 127) / 128) * 128 / 4;
  static constexpr int SMEM = S * STAGE_FLOATS * 4 + 4 * T2_YF4 * 16 + 2 * S * 8 + 2 * S * 4 + 256;
};

template <int S>
__global__ void __launch_bounds__(NCONS + 32, 2)
    k2t_sweep(const __grid_constant__ StencilParams p, const __grid_constant__ CUtensorMap tmap, float* out, int ntx,
              int nty, int zc, int nchunk) {
  using C = CfgT2<S>;
  constexpr int SF4 = C::STAGE_FLOATS / 4;
  constexpr int BX4 = BX / 4;
  constexpr int TX4 = TX / 4;
  extern __shared__ __align__(128) float4 dsm4[];
  float4* ysm = dsm4 + S * SF4;                                   // 4 X_{t+1} slots
  uint64_t* full = reinterpret_cast<uint64_t*>(ysm + 4 * T2_YF4);
  uint64_t* empty = full + S;
  int* stage_item = reinterpret_cast<int*>(empty + S);
  int* slot_sm = stage_item + S;

  const int ntile = ntx * nty;
  const int nitems = ntile * nchunk;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  if (threadIdx.x == 0) {
    for (int s = 0; s < S; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NW);
    }
    fence_mbar_init();
    *slot_sm = claim_launch_slot(g_launch);
  }
  __syncthreads();
  const int slot = *slot_sm;
  pdl_launch_dependents();   // PDL: let the next launch ramp up now
  pdl_wait();                // ... and wait for the previous one before any global access

  if (warp == NW) {
    if (lane == 0) {
      prefetch_tmap(&tmap);
      int s = 0;
      uint32_t pass = 0;
      while (true) {
        const int item = (int)atomicAdd(&g_launch[slot].c[0], 1u);
        const bool done = item >= nitems;
        int nload = 1, x0 = 0, y0 = 0;
        int64_t zs = 0;
        if (!done) {
          const int chunk = item / ntile, tile = item % ntile;
          x0 = (tile % ntx) * T2_TXO;
          y0 = (tile / ntx) * T2_TYO;
          zs = p.reg0 + (int64_t)chunk * zc;
          nload = (int)(min(zs + (int64_t)zc, p.reg1) - zs) + 4;   // X planes zs-2 .. ze+1
        }
        for (int i = 0; i < nload; ++i) {
          if (pass > 0) mbar_wait(&empty[s], (pass - 1) & 1);
          if (i == 0) stage_item[s] = done ? -1 : item;
          if (!done) {
            const int64_t lz = plane_of(p, p.z_off + zs - 2 + i);   // never constant (no CONSTANT kind here)
            mbar_arrive_expect_tx(&full[s], C::TX_BYTES);
            tma_load_3d(dsm4 + s * SF4, &tmap, &full[s], x0 - 8, y0 - 2, (int)lz);
          } else {
            mbar_arrive(&full[s]);
          }
          if (++s == S) { s = 0; ++pass; }
        }
        if (done) break;
      }
    }
  } else {
    const int nx = (int)p.n[2], ny = (int)p.n[1];
    const int kx = p.kind[2], ky = p.kind[1], kz = p.kind[0];
    const int gnz = (int)p.gnz;
    const int rsx = (int)pad_remap(-1, nx, kx);                        // source column of x = -1
    const int rex = (int)(pad_remap(nx, nx, kx) - (nx - 4));           // element of x = nx in the last float4
    int sn = 0;
    uint32_t pn = 0;
    while (true) {
      mbar_wait(&full[sn], pn & 1);
      const int item = stage_item[sn];
      if (item < 0) {
        __syncwarp();
        if (lane == 0) mbar_arrive(&empty[sn]);
        break;
      }
      named_bar_sync(1, NCONS);     // previous item's readers are done with the X_{t+1} ring
      const int chunk = item / ntile, tile = item % ntile;
      const int x0 = (tile % ntx) * T2_TXO, y0 = (tile / ntx) * T2_TYO;
      const int64_t zs = p.reg0 + (int64_t)chunk * zc;
      const int nzc = (int)(min(zs + (int64_t)zc, p.reg1) - zs);
      const int xo = x0 - 4 + 4 * lane;                 // this lane's X_{t+1} / output columns
      const bool pl = xo == 0, pr = xo + 4 == nx;       // x-halo out of grid for this lane
      // (clamp / mirror / reflect: the x = -1 / nx tap is one of the lane's
      // own 4 values; a float4 element index, resolved by selects)
      // X rows (box origin y0-2) and X_{t+1} rows (tile origin y0-1) of this
      // warp's two rows, with the pad redirect folded into the row offsets
      int xm[2], xq[2], ym_[2], yq[2];
#pragma unroll
      for (int jj = 0; jj < 2; ++jj) {
        const int rr = warp * 2 + jj, gy = y0 - 1 + rr;
        xm[jj] = -BX4;
        xq[jj] = BX4;
        if (gy - 1 < 0) xm[jj] = (min(max((int)pad_remap(gy - 1, ny, ky) - (y0 - 2), 0), T2_BY - 1) - (rr + 1)) * BX4;
        if (gy + 1 >= ny) xq[jj] = (min(max((int)pad_remap(gy + 1, ny, ky) - (y0 - 2), 0), T2_BY - 1) - (rr + 1)) * BX4;
        ym_[jj] = -TX4;
        yq[jj] = TX4;
        if (gy - 1 < 0) ym_[jj] = (min(max((int)pad_remap(gy - 1, ny, ky) - (y0 - 1), 0), T2_TY - 1) - rr) * TX4;
        if (gy + 1 >= ny) yq[jj] = (min(max((int)pad_remap(gy + 1, ny, ky) - (y0 - 1), 0), T2_TY - 1) - rr) * TX4;
        if (rr == 0) ym_[jj] = 0;                  // rows 0 and 15 produce no output: stay in the slot
        if (rr == T2_TY - 1) yq[jj] = 0;
      }
      int xst[3];                // stages of X planes yz-1, yz, yz+1
      int yslot[3];              // X_{t+1} ring slots of planes oz-1, oz, oz+1
      // warm-up: X planes zs-2, zs-1
      for (int k = 0; k < 2; ++k) {
        if (k > 0) mbar_wait(&full[sn], pn & 1);
        xst[k] = sn;
        if (++sn == S) { sn = 0; ++pn; }
      }
      // Y plane i (global zs-1+i) lives in slot i & 3; remember which are real
      int yreal[3] = {-1, -1, -1};
      for (int i = 0; i < nzc + 2; ++i) {
        const int yz = (int)(p.z_off + zs) - 1 + i;     // global plane of X_{t+1}
        mbar_wait(&full[sn], pn & 1);
        xst[2] = sn;
        if (++sn == S) { sn = 0; ++pn; }
        const int ys = i & 3;
        const bool inside = yz >= 0 && yz < gnz;
        {
          // ---- step 1: X_{t+1} plane yz on the extended tile (computed for a
          // plane outside the grid too — from the producer's remapped planes —
          // and never read: its slot is aliased away below; no branch) ----
#pragma unroll
          for (int jj = 0; jj < 2; ++jj) {
            const int rr = warp * 2 + jj;
            const int rb = (rr + 1) * BX4 + 1 + lane;    // X box row of y, centre float4 of the lane
            const int cb = xst[1] * SF4;
            const float4 c = dsm4[cb + rb];
            const float4 e = dsm4[cb + (rr + 1) * BX4 + (lane == 0 ? 0 : (TX + XH) / 4)];
            float l = __shfl_up_sync(FULL, c.w, 1);
            float r = __shfl_down_sync(FULL, c.x, 1);
            if (lane == 0) l = e.w;
            if (lane == 31) r = e.x;
            if (pl) l = pick4(rsx, c, 0.0f);
            if (pr) r = pick4(rex, c, 0.0f);
            Win<1> w;
            w.x[0] = l; w.x[1] = c.x; w.x[2] = c.y; w.x[3] = c.z; w.x[4] = c.w; w.x[5] = r;
            set4(w.ym[0], dsm4[cb + rb + xm[jj]]);
            set4(w.yp[0], dsm4[cb + rb + xq[jj]]);
            set4(w.zm[0], dsm4[xst[0] * SF4 + rb]);
            set4(w.zp[0], dsm4[xst[2] * SF4 + rb]);
            const float4 pw = make_float4(0.f, 0.f, 0.f, 0.f);
            float4 v;
            v.x = eval<K2_WSTAR, 1, 0>(p, w, pw, 0, 0, 0);
            v.y = eval<K2_WSTAR, 1, 1>(p, w, pw, 0, 0, 0);
            v.z = eval<K2_WSTAR, 1, 2>(p, w, pw, 0, 0, 0);
            v.w = eval<K2_WSTAR, 1, 3>(p, w, pw, 0, 0, 0);
            ysm[ys * T2_YF4 + rr * TX4 + lane] = v;
          }
        }
        // X plane yz-1 is done
        __syncwarp();
        if (lane == 0) mbar_arrive(&empty[xst[0]]);
        xst[0] = xst[1];
        xst[1] = xst[2];
        yreal[0] = yreal[1];
        yreal[1] = yreal[2];
        yreal[2] = inside ? ys : -1;
        named_bar_sync(1, NCONS);
        if (i < 2) continue;
        // ---- step 2: X_{t+2} plane oz = yz - 1 from X_{t+1} planes oz-1..oz+1 ----
        const int oz = yz - 1;
        // ring slots with the pad of X_{t+1} in z (a plane outside the grid
        // aliases the remapped plane, which is one of the three); interior
        // planes (all but the first and last of the grid) take the fast path
        if (oz >= 1 && oz + 1 < gnz) {
          yslot[0] = yreal[0];
          yslot[1] = yreal[1];
          yslot[2] = yreal[2];
        } else {
#pragma unroll
          for (int k = 0; k < 3; ++k) {
            const int gzk = oz - 1 + k;
            int src = k;
            if (gzk < 0 || gzk >= gnz) src = (int)pad_remap(gzk, gnz, kz) - (oz - 1);
            yslot[k] = (src == 0 ? yreal[0] : (src == 1 ? yreal[1] : yreal[2]));
          }
        }
        float* op = out + ((int64_t)(oz - p.z_off) + p.ghost) * p.plane;
#pragma unroll
        for (int jj = 0; jj < 2; ++jj) {
          const int rr = warp * 2 + jj, gy = y0 - 1 + rr;
          const int rb = rr * TX4 + lane;
          const float4 c = ysm[yslot[1] * T2_YF4 + rb];
          float l = __shfl_up_sync(FULL, c.w, 1);
          float r = __shfl_down_sync(FULL, c.x, 1);
          if (pl) l = pick4(rsx, c, 0.0f);
          if (pr) r = pick4(rex, c, 0.0f);
          Win<1> w;
          w.x[0] = l; w.x[1] = c.x; w.x[2] = c.y; w.x[3] = c.z; w.x[4] = c.w; w.x[5] = r;
          set4(w.ym[0], ysm[yslot[1] * T2_YF4 + rb + ym_[jj]]);
          set4(w.yp[0], ysm[yslot[1] * T2_YF4 + rb + yq[jj]]);
          set4(w.zm[0], ysm[yslot[0] * T2_YF4 + rb]);
          set4(w.zp[0], ysm[yslot[2] * T2_YF4 + rb]);
          const float4 pw = make_float4(0.f, 0.f, 0.f, 0.f);
          float4 v;
          v.x = eval<K2_WSTAR, 1, 0>(p, w, pw, 0, 0, 0);
          v.y = eval<K2_WSTAR, 1, 1>(p, w, pw, 0, 0, 0);
          v.z = eval<K2_WSTAR, 1, 2>(p, w, pw, 0, 0, 0);
          v.w = eval<K2_WSTAR, 1, 3>(p, w, pw, 0, 0, 0);
          const bool ok = lane >= 1 && lane <= 30 && rr >= 1 && rr <= T2_TYO && xo < nx && gy < ny;
          if (ok) stg128(op + (int64_t)gy * nx + xo, v);
        }
      }
      // the chunk's last two X planes are still held
      __syncwarp();
      if (lane == 0) {
        mbar_arrive(&empty[xst[0]]);
        mbar_arrive(&empty[xst[1]]);
      }
    }
  }
  __syncthreads();
  if (threadIdx.x == 0) {
    __threadfence();
    const unsigned prev = atomicAdd(&g_launch[slot].c[1], 1u);
    if (prev == gridDim.x - 1) {
      release_launch_slot(g_launch, slot);
    }
  }
}

// ---------------------------------------------------------------------------
// host side
// ---------------------------------------------------------------------------
bool star_weights(const StencilParams& p, int R) {
  const int S = 2 * R + 1;
  for (int kz = 0; kz < S; ++kz)
    for (int ky = 0; ky < S; ++ky)
      for (int kx = 0; kx < S; ++kx) {
        const int nax = (kz != R) + (ky != R) + (kx != R);
        if (nax > 1 && p.wbox[(kz * S + ky) * S + kx] != 0.0f) return false;
      }
  return true;
}

struct Launcher {
  const void* fn;
  int smem;
  int ty;
  int ctas_per_sm;
};

template <int OP, int R, int RPW, int S, bool ZC, bool FZ, int PSN>
Launcher get_launcher() {
  static Launcher L{};
  static std::once_flag once;
  std::call_once(once, [] {
    using C = Cfg<R, RPW, S, (OP == K2_HOTSPOT || OP == K2_ACOUSTIC) ? PSN : 0>;
    auto fn = k2_sweep<OP, R, RPW, S, ZC, FZ, PSN>;
    cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, C::SMEM);
    int occ = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, fn, NCONS + 32, C::SMEM) != cudaSuccess) occ = 1;
    cudaGetLastError();
    L = Launcher{reinterpret_cast<const void*>(fn), C::SMEM, C::TY, occ > 0 ? occ : 1};
  });
  return L;
}

template <int OP, int R, int RPW, int S, int PSN = 3>
Launcher get_launcher_zf(bool zc, bool fz) {
  if (fz) return zc ? get_launcher<OP, R, RPW, S, true, true, PSN>() : get_launcher<OP, R, RPW, S, false, true, PSN>();
  return zc ? get_launcher<OP, R, RPW, S, true, false, PSN>() : get_launcher<OP, R, RPW, S, false, false, PSN>();
}

Launcher pick(const StencilParams& p) {
  const int R = p.radius;
  // non-zero value-pad planes in z are possible (zero ones are TMA out-of-bounds fills)
  const bool zc = p.kind[0] == PAD_CONSTANT && p.pad_value != 0.0f;
  const bool fz = p.put_lo || p.put_hi || p.fused_step || p.wait_lo || p.wait_hi;   // fused halo launch
  if (p.op == OP_WEIGHTED) {
    if (R == 1 && !star_weights(p, 1)) {
      bool corners = false;
      for (int kz = 0; kz < 3; kz += 2)
        for (int ky = 0; ky < 3; ky += 2)
          for (int kx = 0; kx < 3; kx += 2) corners |= p.wbox[(kz * 3 + ky) * 3 + kx] != 0.0f;
      if (!corners) {
        const char* eb = getenv("LIFT_K2_BOX");      // A/B: (rows per warp, stages)
        if (eb && atoi(eb) == 1) return get_launcher_zf<K2_WBOX19, 1, 1, 8, 0>(zc, fz);
        if (eb && atoi(eb) == 2) return get_launcher_zf<K2_WBOX19, 1, 3, 6, 0>(zc, fz);
        return get_launcher_zf<K2_WBOX19, 1, 2, 7, 0>(zc, fz);
      }
      return get_launcher_zf<K2_WBOX, 1, 2, 7, 0>(zc, fz);
    }
    if (R == 1) return get_launcher_zf<K2_WSTAR, 1, 2, 7, 0>(zc, fz);
    const char* e2 = getenv("LIFT_K2_R2");            // A/B: (rows per warp, stages)
    if (e2 && atoi(e2) == 1) return get_launcher_zf<K2_WSTAR, 2, 1, 8, 0>(zc, fz);
    if (e2 && atoi(e2) == 2) return get_launcher_zf<K2_WSTAR, 2, 3, 6, 0>(zc, fz);
    return get_launcher_zf<K2_WSTAR, 2, 2, 8, 0>(zc, fz);
  }
  // the point-wise grid's TMA ring was the top stall of Acoustic-13 (16.6% of
  // samples waiting on it with 3 slots): radius 1 takes 5 slots (Acoustic-7
  // 484 -> 506, Hotspot3D 276 -> 305 Gpts/s).  LIFT_K2_PW=1: the round-1
  // (S, 3) rings.  (Reading it with global loads two planes ahead instead of
  // a ring measured 20% slower: register spills.)
  const char* e = getenv("LIFT_K2_PW");
  const int pv = e ? atoi(e) : 0;
  if (p.op == OP_HOTSPOT3D) {
    if (pv == 1) return get_launcher_zf<K2_HOTSPOT, 1, 2, 5, 3>(zc, fz);
    const char* eh = getenv("LIFT_K2_HS");          // A/B: small-nz column shapes
    const int hs = eh ? atoi(eh) : 0;
    if (hs == 1) return get_launcher_zf<K2_HOTSPOT, 1, 1, 10, 8>(zc, fz);
    if (hs == 2) return get_launcher_zf<K2_HOTSPOT, 1, 1, 12, 8>(zc, fz);
    if (hs == 3) return get_launcher_zf<K2_HOTSPOT, 1, 2, 10, 8>(zc, fz);
    if (hs == 4) return get_launcher_zf<K2_HOTSPOT, 1, 1, 6, 6>(zc, fz);
    return get_launcher_zf<K2_HOTSPOT, 1, 2, 5, 5>(zc, fz);
  }
  if (R == 1) {
    if (pv == 1) return get_launcher_zf<K2_ACOUSTIC, 1, 2, 5, 3>(zc, fz);
    return get_launcher_zf<K2_ACOUSTIC, 1, 2, 5, 5>(zc, fz);
  }
  // radius 2: the 5 live planes need a deep plane ring too; (7 plane stages,
  // 4 point-wise slots) fits 2 CTAs per SM (Acoustic-13 1024^3: 451 Gpts/s
  // vs 448 for (8, 3) and 411 for (6, 5); 8-row tiles at 3 CTAs/SM and
  // 24-row tiles measured 379 / 371 vs 466, profiles/r01_sweep_acoustic13_shapes.txt)
  if (pv == 1) return get_launcher_zf<K2_ACOUSTIC, 2, 2, 8, 3>(zc, fz);
  return get_launcher_zf<K2_ACOUSTIC, 2, 2, 7, 4>(zc, fz);
}

struct MapEntry {
  const float* base;
  int64_t nx, ny, nz;
  int bx, by;
  CUtensorMap map;
};

bool get_map(const float* base, int64_t nx, int64_t ny, int64_t nz, int bx, int by, CUtensorMap* out,
             std::string* err) {
  thread_local MapEntry cache[8];
  thread_local int next = 0;
  for (auto& e : cache)
    if (e.base == base && e.nx == nx && e.ny == ny && e.nz == nz && e.bx == bx && e.by == by) {
      *out = e.map;
      return true;
    }
  MapEntry e{base, nx, ny, nz, bx, by, {}};
  if (!encode_tensor_map_3d(&e.map, base, nx, ny, nz, (uint32_t)bx, (uint32_t)by, 1, err)) return false;
  cache[next] = e;
  next = (next + 1) % 8;
  *out = e.map;
  return true;
}


}  // namespace

bool sweep3d_supported(const StencilParams& p) {
  if (has_dampen(p)) return false;     // DAMPEN pads run on K5 / K0
  const int R = p.radius;
  if (R != 1 && R != 2) return false;
  for (int d = 0; d < 3; ++d)
    if (p.size[d] != 2 * R + 1 || p.lo[d] != R || p.hi[d] != R || p.step[d] != 1) return false;
  if (p.op == OP_WEIGHTED) {
    if (!star_weights(p, R) && R != 1) return false;      // 3x3x3 boxes run on K2_WBOX
  } else if (p.op == OP_HOTSPOT3D) {
    if (R != 1) return false;
  } else if (p.op != OP_ACOUSTIC) {
    return false;
  }
  if (p.n[2] % 4 != 0) return false;
  if (p.n[2] * p.n[1] >= (1ll << 31) || p.gnz >= (1ll << 31) || p.n[0] + 2 * p.ghost >= (1ll << 31)) return false;
  return true;
}

cudaError_t launch_sweep3d(const StencilParams& p, const float* in0, const float* in1, float* out,
                           cudaStream_t stream, int num_sms, std::string* err) {
  const int64_t nz_reg = p.reg1 - p.reg0;
  if (nz_reg <= 0) return cudaSuccess;
  if (column3d_supported(p, in0, in1)) return launch_column3d(p, in0, in1, out, stream, err);
  const Launcher L = pick(p);
  const int R = p.radius;
  const float* slid = (p.op == OP_ACOUSTIC) ? in1 : in0;
  const float* pw = (p.op == OP_ACOUSTIC) ? in0 : (p.op == OP_HOTSPOT3D ? in1 : nullptr);
  CUtensorMap map, pwmap;
  if (!get_map(slid, p.n[2], p.n[1], p.n[0] + 2 * p.ghost, BX, L.ty + 2 * R, &map, err)) return cudaErrorInvalidValue;
  if (pw) {
    if (!get_map(pw, p.n[2], p.n[1], p.n[0] + 2 * p.ghost, TX, L.ty, &pwmap, err)) return cudaErrorInvalidValue;
  } else {
    pwmap = map;
  }
  const int ntx = (int)((p.n[2] + TX - 1) / TX);
  const int nty = (int)((p.n[1] + L.ty - 1) / L.ty);
  const int64_t tiles = (int64_t)ntx * nty;
  const int64_t slots = (int64_t)num_sms * L.ctas_per_sm;
  // z-chunk: ~8 items per CTA for dynamic balance, at least 16 planes (halo
  // re-load <= 2R/16) — unless the grid is too small to give every CTA two
  // items (e.g. Hotspot3D's 8 planes), then parallelism wins over halo reuse
  const int64_t work = nz_reg * tiles;
  int64_t zc = (work + 8 * slots - 1) / (8 * slots);
  const int64_t zmin = std::min<int64_t>(16, std::max<int64_t>(2, (work + 2 * slots - 1) / (2 * slots)));
  if (zc < zmin) zc = zmin;
  if (work < 16 * slots) {
    // small (L2-resident, latency-bound) grids, e.g. Hotspot3D's 8 planes: the
    // step takes about (waves of items) x (planes loaded per item), so pick
    // the chunk that minimises ceil(items / slots) * (zc + 2R)
    int64_t best = -1;
    for (int64_t z = 1; z <= nz_reg; ++z) {
      const int64_t it = tiles * ((nz_reg + z - 1) / z);
      const int64_t cost = ((it + slots - 1) / slots) * (z + 2 * R);
      if (best < 0 || cost < best) {
        best = cost;
        zc = z;
      }
    }
  }
  // Large grids, measured per kernel family (profiles/r01_sweep_zchunk.txt):
  // the memory-bound radius-1 sweeps (7-point weighted star, Acoustic-7) run
  // fastest with short chunks — CTAs in flight then stay within a narrow z
  // window (halo planes and rows are L2 hits) and the launch's tail is short:
  // J3D7 512^3 766 -> 825 Gpts/s at 6 planes (~20 planes' worth of items in
  // flight for the weighted star, ~40 for Acoustic, whose items carry a
  // point-wise grid); the instruction-heavier radius-2 and box sweeps keep
  // long chunks (their 2R warm-up planes per chunk cost issue slots) and only
  // shorten the chunks of the last waves (guided tail).
  int64_t tail_zc = 0;
  if (work >= 16 * slots) {
    const bool box = p.op == OP_WEIGHTED && !star_weights(p, 1);
    if (R == 1 && !box && (p.op == OP_WEIGHTED || p.op == OP_ACOUSTIC)) {
      const int64_t k = p.op == OP_ACOUSTIC ? 40 : 20;
      zc = std::min<int64_t>(64, std::max<int64_t>(4, (k * tiles + slots / 2) / slots));
    } else if (!p.fused_step) {       // (the fused step keeps uniform chunks: boundary chunks first)
      tail_zc = p.op == OP_ACOUSTIC ? 16 : 8;
    }
  }
  if (const char* e = getenv("LIFT_K2_ZC")) zc = std::max<int64_t>(1, atoll(e));   // tuning hook
  if (p.fused_step && zc < p.ghost) zc = p.ghost;     // boundary planes stay in the first / last chunk
  if (zc > nz_reg) zc = nz_reg;
  int64_t nchunk = (nz_reg + zc - 1) / zc;
  // guided tail: the last ~tailw waves of items take zc2-plane chunks
  int64_t n1 = nchunk, zc2 = zc;
  {
    const char* e2 = getenv("LIFT_K2_ZC2");
    const char* ew = getenv("LIFT_K2_TAILW");
    const int64_t want = e2 ? atoll(e2) : tail_zc;
    const int64_t tailw = ew ? std::max<int64_t>(1, atoll(ew)) : 2;
    if (want > 0 && want < zc && !p.fused_step && work >= 16 * slots) {
      const int64_t nsmall = (tailw * slots + tiles - 1) / tiles;      // small chunks per tile column
      const int64_t z2 = nsmall * want;
      if (z2 < nz_reg) {
        n1 = (nz_reg - z2) / zc;
        zc2 = want;
        nchunk = n1 + (nz_reg - n1 * zc + zc2 - 1) / zc2;
      }
    }
  }
  const int64_t items = tiles * nchunk;
  if (items > 0x7fffffff) return cudaErrorInvalidConfiguration;
  int64_t grid = slots < items ? slots : items;
  int ntx_i = ntx, nty_i = nty, zc_i = (int)zc, nch_i = (int)nchunk, n1_i = (int)n1, zc2_i = (int)zc2;
  void* args[] = {(void*)&p, (void*)&map, (void*)&pwmap, (void*)&slid, (void*)&out,
                  &ntx_i, &nty_i, &zc_i, &nch_i, &n1_i, &zc2_i};
  const bool fz = p.put_lo || p.put_hi || p.fused_step || p.wait_lo || p.wait_hi;
  // PDL for the fused halo launches is an A/B knob (LIFT_FUSED_PDL=1): the
  // kernel's flag spins come after its griddepcontrol.wait, so a dependent
  // launch cannot run ahead of the step it depends on
  static const bool fused_pdl = [] {
    const char* e = getenv("LIFT_FUSED_PDL");
    return e && e[0] == '1';
  }();
  set_last_kernel("k2_sweep");
  return launch_kernel(L.fn, dim3((unsigned)grid), dim3(NCONS + 32), args, (size_t)L.smem, stream, !fz || fused_pdl);
}

}  // namespace lift

namespace lift {

bool sweep3d_t2_supported(const StencilParams& p) {
  if (p.op != OP_WEIGHTED || p.radius != 1 || !sweep3d_supported(p)) return false;
  if (!star_weights(p, 1)) return false;
  for (int d = 0; d < 3; ++d)
    if (p.kind[d] != PAD_CLAMP && p.kind[d] != PAD_MIRROR && p.kind[d] != PAD_REFLECT) return false;
  if (p.put_lo || p.put_hi || p.fused_step) return false;
  if (p.slab && p.ghost < 2) return false;        // X_{t+1} of the planes next to the slab edge
  return true;
}

cudaError_t launch_sweep3d_t2(const StencilParams& p, const float* in, float* out, cudaStream_t stream, int num_sms,
                              std::string* err) {
  if (sweep3d_r2_supported(p)) return launch_sweep3d_r2(p, in, out, stream, num_sms, err);
  const int64_t nz_reg = p.reg1 - p.reg0;
  if (nz_reg <= 0) return cudaSuccess;
  constexpr int S = 5;
  static Launcher L{};
  static std::once_flag once;
  std::call_once(once, [] {
    auto fn = k2t_sweep<S>;
    cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, CfgT2<S>::SMEM);
    int occ = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, fn, NCONS + 32, CfgT2<S>::SMEM) != cudaSuccess) occ = 1;
    cudaGetLastError();
    L = Launcher{reinterpret_cast<const void*>(fn), CfgT2<S>::SMEM, T2_TYO, occ > 0 ? occ : 1};
  });
  CUtensorMap map;
  if (!get_map(in, p.n[2], p.n[1], p.n[0] + 2 * p.ghost, BX, T2_BY, &map, err)) return cudaErrorInvalidValue;
  const int ntx = (int)((p.n[2] + T2_TXO - 1) / T2_TXO);
  const int nty = (int)((p.n[1] + T2_TYO - 1) / T2_TYO);
  const int64_t tiles = (int64_t)ntx * nty;
  const int64_t slots = (int64_t)num_sms * L.ctas_per_sm;
  const int64_t work = nz_reg * tiles;
  int64_t zc = (work + 8 * slots - 1) / (8 * slots);
  const int64_t zmin = std::min<int64_t>(16, std::max<int64_t>(2, (work + 2 * slots - 1) / (2 * slots)));
  if (zc < zmin) zc = zmin;
  if (zc > nz_reg) zc = nz_reg;
  const int64_t nchunk = (nz_reg + zc - 1) / zc;
  const int64_t items = tiles * nchunk;
  if (items > 0x7fffffff) return cudaErrorInvalidConfiguration;
  int64_t grid = slots < items ? slots : items;
  int ntx_i = ntx, nty_i = nty, zc_i = (int)zc, nch_i = (int)nchunk;
  void* args[] = {(void*)&p, (void*)&map, (void*)&out, &ntx_i, &nty_i, &zc_i, &nch_i};
  set_last_kernel("k2t_sweep");
  return launch_kernel(L.fn, dim3((unsigned)grid), dim3(NCONS + 32), args, (size_t)L.smem, stream, true);
}

}  // namespace lift
