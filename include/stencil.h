/*
 * stencil.h — C ABI of the B200 Lift-stencil hot path.
 *
 * The operation is the paper's problem statement (§3.4):
 *
 *     out = map_n(f, slide_n(size, step, pad_n(l, r, h, input)))
 *
 *   pad  grows each dimension d by l_d on the left and r_d on
 *                       the right; padded index j reads input[h_d(j - l_d, n_d)]
 *                       (reindexing variant) or the constant pad_value
 *                       (value variant).  h may differ per dimension.
 *   slide  (P:467-479,  window o is padded indices o*step + k, k in [0,size);
 *           P:567-630)  o_d in [0, floor((n_d + l_d + r_d - size_d)/step_d) + 1).
 *   map  f is applied to every window; extra grids are zipped
 *                       point-wise (zip; Listing 3).
 *   iterate     repeats the step, feeding the output back.
 *
 * Conventions (all functions):
 *   - grids are contiguous fp32, row-major, extents slowest-first
 *     (``[[T]_m]_n`` has n outermost); ndim in {1, 2, 3};
 *   - every grid pointer passed to apply/iterate is a DEVICE pointer owned by
 *     the caller; weights/params are HOST pointers copied into the plan;
 *   - ``stream`` is a cudaStream_t passed as void* (NULL = legacy default
 *     stream); apply/apply_region/iterate are asynchronous, stream-ordered,
 *     allocate nothing and are CUDA-graph capturable;
 *   - every function returns a stencil_status; nothing aborts and no C++
 *     exception crosses the ABI; stencil_last_error() gives a thread-local
 *     message for the last failure.  Asynchronous kernel faults surface at the
 *     caller's next synchronisation, as with any CUDA library.
 *   - there is no CPU fallback: without a usable CUDA device every call that
 *     launches work returns STENCIL_E_CUDA.
 */
#ifndef LIFT_STENCIL_H
#define LIFT_STENCIL_H

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef struct stencil_plan_s* stencil_plan;   /* opaque, owned by the library */

typedef enum {
  STENCIL_OK = 0,
  STENCIL_E_INVALID = 1,      /* argument violates the pad/slide/map types  */
  STENCIL_E_UNSUPPORTED = 2,  /* valid, but not built (e.g. ndim > 3)        */
  STENCIL_E_CUDA = 3,         /* a CUDA call or launch failed               */
  STENCIL_E_NOMEM = 4
} stencil_status;

/* Boundary index functions h of pad (A1-A5). */
typedef enum {
  STENCIL_PAD_CLAMP = 0,      /* (i<0) ? 0 : ((i>=n) ? n-1 : i) */
  STENCIL_PAD_MIRROR = 1,     /* symmetric, edge repeated (numpy 'symmetric')  A2 */
  STENCIL_PAD_WRAP = 2,       /* ((i mod n) + n) mod n                         A3 */
  STENCIL_PAD_CONSTANT = 3,   /* value variant of pad: pad_value              A4 */
  STENCIL_PAD_REFLECT = 4,    /* edge not repeated (numpy 'reflect')          A2 */
  STENCIL_PAD_DAMPEN = 5      /* "dampening boundary conditions where the
                                 out-of-bound value decreases with the distance
                                 to the boundary", reading A29: the
                                 cell d steps outside holds the nearest element
                                 times decay^d (stencil_plan_set_pad_decay);
                                 WEIGHTED only; decay 1 = CLAMP, 0 = zeros    */
} stencil_pad;

/* Neighbourhood functions f of map (A13-A20). */
typedef enum {
  STENCIL_OP_WEIGHTED = 0,   /* sum_k w_k W[k], taps in row-major order; 1 input   */
  STENCIL_OP_HOTSPOT3D = 1,  /* Rodinia hotspot3D (A16): inputs {T (slid), P};
                                params {cc,cn,cs,ce,cw,ct,cb,sdc,amb}; 3D, size 3  */
  STENCIL_OP_SRAD1 = 2,      /* Rodinia SRAD kernel 1 (A18): input {I} -> c;
                                params {q0sqr}; 2D, size 3                         */
  STENCIL_OP_SRAD2 = 3,      /* Rodinia SRAD kernel 2 (A18): inputs {c, I} -> I';
                                params {lambda}; 2D, size 3                        */
  STENCIL_OP_ACOUSTIC = 4,   /* Listing 3 (A19/A20): inputs {prev
                                (point-wise), cur (slid)} -> next; params
                                {lambda^2, loss1, loss2}; 3D, size 3 (7-pt) or
                                5 (13-pt); ``out`` may alias ``prev``              */
  STENCIL_OP_HOTSPOT2D = 5,  /* Rodinia hotspot (A26, Table 1): inputs {T
                                (slid), P (point-wise)}; params {step/Cap, 1/Rx,
                                1/Ry, 1/Rz, amb}; 2D, size 3                       */
  STENCIL_OP_GRADIENT = 6,   /* Rawat et al. 2D gradient (A25, Table 1):
                                I + 1/sqrt(eps + sum of squared differences to
                                the 4 neighbours); params {eps}; 2D, size 3        */
  STENCIL_OP_SRAD = 7        /* one full SRAD iteration (A27, NEXT-2): q0^2 =
                                var/mean^2 of the input (fp64 reduction on the
                                device), c = SRAD1, I' = SRAD2 fused in one pass;
                                input {I}; params {lambda}; 2D, size 3, reindexing
                                pads; the plan owns a small device workspace      */
} stencil_op;

/* Which kernel family executes a plan (stencil_plan_variant). */
typedef enum {
  STENCIL_VARIANT_AUTO = -1,
  STENCIL_VARIANT_GENERIC = 0,   /* K0: one thread per output, remapped loads  */
  STENCIL_VARIANT_TILE2D = 1,    /* K1: TMA halo tile, 2D                       */
  STENCIL_VARIANT_SWEEP3D = 2,   /* K2: TMA plane ring, 2.5D sweep along z      */
  STENCIL_VARIANT_PERSIST3D = 3, /* K4: all n steps of stencil_iterate in one
                                    persistent cooperative launch (small,
                                    L2-resident 3D radius-1 star / Hotspot3D
                                    grids; opt-in with LIFT_K4=1 — measured
                                    slower than K2 steps; reported by
                                    stencil_plan_last_variant, not forceable)  */
  STENCIL_VARIANT_GATHER = 4,    /* K5: WEIGHTED plans the TMA families do not
                                    take (step > 1, even / asymmetric windows,
                                    1D, wide boxes, unaligned 3D) through
                                    shared-memory tiles of the input box        */
  STENCIL_VARIANT_RESIDENT3D = 5 /* K6: all n steps of stencil_iterate for a
                                    few-plane (nz <= 16) 3D radius-1 star /
                                    Hotspot3D grid that fits in the device's
                                    shared memory (one tile per SM), in one
                                    cooperative launch with point-to-point
                                    step flags; opt-in with LIFT_K6=1 (measured
                                    slower than graph-replayed K2C sweeps);
                                    reported by stencil_plan_last_variant, not
                                    forceable                                   */
} stencil_variant;

/*
 * Create a plan for one stencil.
 *   out        : receives the plan handle (NULL on failure).
 *   device     : CUDA device ordinal the plan's launches target.
 *   ndim       : 1, 2 or 3.
 *   extents    : [ndim] input extents n_d, slowest first, each >= 1.
 *   size, step : [ndim] slide(size_d, step_d), each >= 1.
 *   pad_lo/hi  : [ndim] pad(l_d, r_d), each >= 0; n_d + l_d + r_d >= size_d.
 *   kind       : [ndim] stencil_pad per dimension.
 *   pad_value  : value for STENCIL_PAD_CONSTANT dimensions.
 *   op         : stencil_op.
 *   weights    : host, prod(size) floats, row-major over the window (tap k is
 *                padded index o*step + k: cross-correlation, reading A7);
 *                required for WEIGHTED (at most 125 non-zero taps), NULL
 *                otherwise; copied.
 *   params     : host, n_params op constants (see stencil_op); copied.
 * Errors: E_INVALID for any type violation listed above, a wrong op/ndim
 * combination or a NULL weights pointer for WEIGHTED; E_UNSUPPORTED for
 * ndim > 3 or more than 125 non-zero taps.
 */
stencil_status stencil_plan_create(stencil_plan* out, int device, int ndim,
                                   const int64_t* extents, const int32_t* size,
                                   const int32_t* step, const int32_t* pad_lo,
                                   const int32_t* pad_hi, const int32_t* kind,
                                   float pad_value, int32_t op,
                                   const float* weights, const float* params,
                                   int32_t n_params);

/* Output extents o_d = floor((n_d + l_d + r_d - size_d) / step_d) + 1. */
stencil_status stencil_plan_output_extents(stencil_plan plan, int64_t* out_extents);

/*
 * Slab mode (multi-GPU decomposition along dimension 0, 3D plans only).
 * The plan's extents are the OWNED slab (n0_local, n1, n2) of a global grid
 * with n0 = global_n0 planes; the slab's first owned plane is global plane
 * z_offset.  Every grid buffer passed to apply/iterate then holds
 * n0_local + 2*ghost planes: ghost planes [0, ghost) precede the owned planes
 * and [ghost + n0_local, n0_local + 2*ghost) follow them; pointers point at
 * plane 0 of the allocation.  Output planes are written at the same offsets
 * (owned planes only).  Planes outside the global domain are handled by pad
 * against the GLOBAL extent; WRAP in dimension 0 reads the ghost planes (the
 * caller fills them from the ring neighbour).  ghost >= max(pad_lo[0],
 * pad_hi[0]); requires step[0] == 1 and output extents == input extents.
 */
stencil_status stencil_plan_set_slab(stencil_plan plan, int64_t z_offset,
                                     int64_t global_n0, int32_t ghost);

/* Temporal blocking for stencil_iterate (overlapped tiling
 * applied to iterate): steps = 2 lets iterate
 * advance two time steps per pass over HBM where a two-step kernel applies
 * (WEIGHTED 7-point star; K2R with X_{t+1} in registers for x/y CLAMP /
 * MIRROR / REFLECT and z CLAMP / MIRROR, else the shared-memory K2T for z
 * REFLECT); the result is bitwise identical to single steps (an odd step
 * count ends with one single step).  1 forces one step per pass.  0 (the
 * default, AUTO) takes two steps per pass where K2R applies and the grid
 * fills the GPU (>= 8 tiles of 128 x 48 per plane with >= 0.9 useful columns
 * and >= 2048 (plane, tile) pairs; J3D7 512^3: ~1.6x the single-step rate,
 * 256^3: 1.2x), and likewise for the 7-point ACOUSTIC update
 * with zero padding where K2RA applies (iterate with four state buffers).  2 also forces K2RA for the 13-point update and K2CT (two
 * Hotspot3D steps per launch of a few-plane grid, nz <= 16, reindexing pads),
 * which measured no faster than single steps and are not in AUTO.  Returns
 * STENCIL_E_INVALID for steps outside 0..2.  stencil_plan_time_block returns
 * the steps per pass iterate will use (1 or 2). */
stencil_status stencil_plan_set_time_block(stencil_plan plan, int32_t steps);
int32_t stencil_plan_time_block(stencil_plan plan);

/* Force a kernel family (tests: tiling independence) or AUTO. E_UNSUPPORTED if
 * the requested family cannot run this plan. */
stencil_status stencil_plan_set_variant(stencil_plan plan, int32_t variant);
/* The family AUTO (or the forced one) selects for the given pointers. */
int32_t stencil_plan_variant(stencil_plan plan);
/* PAD_DAMPEN dimensions: the factor per cell of distance outside the grid,
 * decay in [0, 1] (default 1).  E_INVALID outside that range.  Applies to
 * subsequent launches. */
stencil_status stencil_plan_set_pad_decay(stencil_plan plan, float decay);
/* The family that ran the plan's most recent apply / iterate launch
 * (STENCIL_VARIANT_PERSIST3D after a K4 iterate; GENERIC before any launch). */
int32_t stencil_plan_last_variant(stencil_plan plan);
/* The kernel function of the plan's most recent launch within its family
 * ("k2_sweep", "k2c_column", "k2t_sweep", "k2r_sweep", "k2ra_sweep",
 * "k2ct_column", "k1_tile", "k1_srad_fused",
 * "k3_wsweep", "k5_gather", "k5_gather (TMA)", "k0_generic", "k4_iterate",
 * "k6_resident"; "none" before any launch).  A static string owned by the
 * library. */
const char* stencil_plan_last_kernel(stencil_plan plan);

/*
 * out = map(f, slide(pad(inputs))) — one application.
 *   inputs   : [n_inputs] device pointers (op arity, stencil_op).
 *   out      : device pointer, output extents (slab: allocation layout).
 * Errors: E_INVALID for wrong n_inputs, NULL pointers, or ``out`` aliasing a
 * slid input; E_CUDA on launch failure.
 */
stencil_status stencil_apply(stencil_plan plan, const float* const* inputs,
                             int32_t n_inputs, float* out, void* stream);

/* Same, restricted to output planes [o0_begin, o0_end) of dimension 0
 * (slab interior / boundary split).  Results are bitwise identical to the
 * corresponding planes of stencil_apply.  Slab plans (stencil_plan_set_slab)
 * may extend the region into the ghost planes, o0_begin >= -(ghost -
 * pad_lo[0]) and o0_end <= n0_local + ghost - pad_hi[0]: the redundant
 * overlap compute of deep halos (ghosts of r*k planes exchanged every k
 * steps; P:739-791 overlapped tiling applied in time); output
 * plane z < 0 is written to ghost plane ghost + z of ``out``. */
stencil_status stencil_apply_region(stencil_plan plan, const float* const* inputs,
                                    int32_t n_inputs, float* out, int64_t o0_begin,
                                    int64_t o0_end, void* stream);

/* TWO time steps of a WEIGHTED 3D plan in one pass over HBM (the two-step
 * kernels of stencil_plan_set_time_block: K2R, or K2T for z REFLECT) on
 * output planes [o0_begin, o0_end): out = S(S(in)) there, bitwise equal to
 * two stencil_apply_region steps (the first over [o0_begin - pad_lo[0],
 * o0_end + pad_hi[0])).  in: 1 device pointer, out: a different buffer of the
 * same layout, both 16-byte aligned.  Slab plans may reach into the ghosts
 * as far as the first step's input stays inside them: o0_begin >= -(ghost -
 * 2 pad_lo[0]), o0_end <= n0_local + ghost - 2 pad_hi[0] (deep halos with
 * two steps per pass).  E_UNSUPPORTED if no two-step kernel
 * takes the plan (stencil_plan_time_block would return 1 for time block 2);
 * E_INVALID for a region outside those limits, bad pointers or aliasing;
 * E_CUDA on launch failure. */
stencil_status stencil_apply2_region(stencil_plan plan, const float* in, float* out, int64_t o0_begin,
                                     int64_t o0_end, void* stream);

/*
 * Fused halo put (slab mode, 3D plans on the TMA sweep kernel): like
 * stencil_apply_region, and every output plane z < ghost is ALSO stored to
 * put_lo + z*plane, every plane z >= n0_local - ghost to
 * put_hi + (z - (n0_local - ghost))*plane — the neighbour ranks' ghost planes
 * through NVLink peer pointers (NULL = no neighbour on that side).  When all
 * stores are done, the kernel's last CTA makes them visible system-wide and
 * release-stores sig_value to *sig_lo / *sig_hi (the neighbours' flags for
 * this rank; NULL = none).  The region must cover the planes to be put.
 * Errors: E_UNSUPPORTED if the plan does not run on the sweep kernel (the
 * caller then exchanges ghosts with stencil_apply_region + NCCL).
 */
stencil_status stencil_apply_region_put(stencil_plan plan, const float* const* inputs, int32_t n_inputs,
                                        float* out, int64_t o0_begin, int64_t o0_end, float* put_lo,
                                        float* put_hi, uint32_t* sig_lo, uint32_t* sig_hi,
                                        uint32_t sig_value, void* stream);

/*
 * One time step of a slab as ONE launch with the halo exchange fused in:
 * computes all owned output planes; the boundary z-chunks are scheduled first;
 * before loading the ghost planes of the first / last chunk the kernel waits
 * (acquire, system scope) until *wait_lo / *wait_hi >= wait_value (this rank's
 * flags, raised by the neighbours' previous step; NULL = no wait); output planes
 * z < ghost / z >= n0_local - ghost are also stored to put_lo / put_hi as in
 * stencil_apply_region_put, and when the first / last chunk is complete the
 * neighbours' flags *sig_lo / *sig_hi are release-stored with sig_value.
 * Needs a slab plan on the TMA sweep kernel (E_UNSUPPORTED otherwise).
 */
stencil_status stencil_slab_step_fused(stencil_plan plan, const float* const* inputs, int32_t n_inputs,
                                       float* out, float* put_lo, float* put_hi, uint32_t* sig_lo,
                                       uint32_t* sig_hi, uint32_t sig_value, const uint32_t* wait_lo,
                                       const uint32_t* wait_hi, uint32_t wait_value, void* stream);

/* Stream-ordered wait: a one-thread kernel on ``stream`` spins (acquire,
 * system scope) until *sig_a >= value and *sig_b >= value (wrap-around
 * compare; NULL pointers are skipped).  Pairs with stencil_apply_region_put. */
stencil_status stencil_wait_signals(const uint32_t* sig_a, const uint32_t* sig_b, uint32_t value,
                                    void* stream);

/*
 * Bounded halo waits.  Every flag wait of the fused slab path (the producer
 * of stencil_slab_step_fused, the kernel of stencil_wait_signals) gives up
 * after a process-wide timeout instead of spinning forever on a neighbour
 * that died or stalled: it records the fault in a host-visible word and lets
 * the launch finish (its ghost planes are then stale).
 *   stencil_set_wait_timeout_ms : the timeout for subsequent launches; 0 =
 *       wait forever; default 10000 ms (environment LIFT_WAIT_TIMEOUT_MS).
 *   stencil_device_fault : after the caller has synchronised the stream,
 *       returns E_CUDA (detail in stencil_last_error: which neighbour) if a
 *       wait timed out since the last check, and clears the record; OK
 *       otherwise.  stencil_slab_step_fused, stencil_apply_region_put and
 *       stencil_wait_signals also check it on entry and return E_CUDA
 *       without launching.
 */
stencil_status stencil_set_wait_timeout_ms(uint32_t ms);
stencil_status stencil_device_fault(void);

/*
 * iterate(in, f, n_steps) with the state rotation of reading A21:
 *   WEIGHTED  : state {X0, X1}            X_{t+1} = S(X_t), ping-pong
 *   HOTSPOT3D, HOTSPOT2D : state {T0, T1}, aux {P}   T_{t+1} = S(T_t, P)
 *   GRADIENT, SRAD : state {X0, X1}       ping-pong like WEIGHTED
 *     (SRAD: each fused pass also writes the fp64 q0 statistics of the image
 *     it produced to the plan's workspace and the next pass of this call
 *     reduces those instead of re-reading the image; only the first pass
 *     reads X0 once more for its q0)
 *   ACOUSTIC  : state {prev, cur}         next overwrites prev; roles swap
 *     or {prev, cur, spare, spare} (n_state 4, four distinct grids): where
 *     the two-step kernel K2RA applies (zero padding, 7/13-point, not a slab,
 *     time block 0 or 2) each pass reads prev and cur once and writes
 *     u^{n+1} and u^{n+2} into the other pair (16 B per point for two steps
 *     instead of 24), bitwise equal to single steps; an odd remainder runs
 *     one single step.  The grid before the newest is state[*result_index ^ 1].
 * *result_index receives the index into ``state`` holding the newest grid
 * (with two-step passes not necessarily n_steps % 2).  n_state must be 2
 * (ACOUSTIC: 2 or 4), else E_INVALID.
 * Requires output extents == input extents.
 */
stencil_status stencil_iterate(stencil_plan plan, float* const* state, int32_t n_state,
                               const float* const* aux, int32_t n_aux, int32_t n_steps,
                               void* stream, int32_t* result_index);

/*
 * End-to-end entry with HOST buffers (pinned or pageable): copies the state
 * and aux grids host->device into plan-owned device buffers, runs
 * stencil_iterate (n_steps >= 1; n_steps == 1 with a non-iterable op is one
 * stencil_apply), copies the newest grid back to host_out (output extents),
 * and synchronises ``stream``.  The device workspace is allocated on first
 * use, kept by the plan and freed by stencil_plan_destroy.
 */
stencil_status stencil_run_host(stencil_plan plan, const float* const* host_state,
                                int32_t n_state, const float* const* host_aux,
                                int32_t n_aux, int32_t n_steps, float* host_out,
                                void* stream);

/*
 * Batched end-to-end entry: n_jobs independent problems of this plan through
 * one call that overlaps the host->device copy of job j+1 and the
 * device->host copy of job j-1 with the compute of job j (three plan-owned
 * device workspace slots; a copy-in, a compute and a copy-out stream ordered
 * by events; PCIe copies run in both directions at once).  Job j reads
 * host_state[j * n_state + s] (s < n_state) and host_aux[j * n_aux + a] and
 * writes its newest grid to host_out[j] — the same computation as
 * stencil_run_host per job, bitwise.  Host buffers should be pinned for the
 * copies to overlap (pageable ones serialise them).  Synchronous: returns
 * when every output is on the host.  E_INVALID for bad buffers or counts
 * (n_jobs >= 1), else as stencil_run_host.  Device memory: 12 grid-sized
 * buffers (3 slots x 4 grids), allocated on first use, kept by the plan and
 * freed by stencil_plan_destroy.  ACOUSTIC jobs use the four grids of a slot
 * as its state (two steps per pass where K2RA applies).
 */
stencil_status stencil_run_host_batch(stencil_plan plan, const float* const* host_state, int32_t n_state,
                                      const float* const* host_aux, int32_t n_aux, int32_t n_steps,
                                      int32_t n_jobs, float* const* host_out);

/* Frees the plan (host memory and any stencil_run_host workspace).  Safe once
 * the caller has synchronised the plan's in-flight work. */
void stencil_plan_destroy(stencil_plan plan);

const char* stencil_status_string(stencil_status status);
const char* stencil_last_error(void);

/* Library build/version string. */
const char* stencil_version(void);

#ifdef __cplusplus
}
#endif

#endif /* LIFT_STENCIL_H */
