// slots.cuh — per-launch dynamic work counters, claimed by the launch itself.
//
// The persistent kernels (K2, K2T, K3, K4) hand out work items from a ticket
// counter and let their last CTA reset it.  Those counters must belong to ONE
// launch while it runs: two launches sharing them (two graphs replayed
// concurrently on two streams, two plans on two streams) would skip or repeat
// items.  A slot index chosen on the host and baked into a captured graph
// cannot guarantee that, so each launch claims its slot on the device, keyed
// by its grid id (%gridid: the context's temporal launch number — distinct
// for every eager launch and for every kernel node of every instantiated
// graph; replays of ONE executable graph reuse its node ids, but CUDA
// serialises the launches of one executable graph, so they never overlap;
// profiles/r02_gridid_probe.txt): slot = (grid id + 1) mod K.
// Every CTA of the launch computes the same slot; the first one to arrive
// takes ownership (CAS 0 -> id), the last one out zeroes the counters and
// then frees it.  Two launches share a slot only if their ids differ by a
// multiple of K = 65536 while both are still running — and then the later
// one WAITS for the slot to be freed instead of sharing it (the index is a
// pure function of the id, so every CTA of a launch agrees on it; probing
// onward would let two CTAs of one launch pick different slots).
#pragma once
#include <cstdint>

namespace lift {

constexpr int kLaunchSlots = 65536;   // 2 MiB of counters per kernel family

struct alignas(32) LaunchSlot {
  unsigned long long owner;   // grid id + 1 of the launch holding the slot, 0 = free
  unsigned int c[6];          // the kernel's counters (ticket, done, ...)
};

__device__ __forceinline__ unsigned long long grid_id() {
  unsigned long long g;
  asm volatile("mov.u64 %0, %%gridid;" : "=l"(g));
  return g;
}

// Called by one thread per CTA; every CTA of a launch gets the same index.
// ``Slot`` has an ``owner`` word; K (a power of two) entries in ``tab``.
template <int K, class Slot>
__device__ __forceinline__ int claim_slot(Slot* tab) {
  const unsigned long long tag = grid_id() + 1ull;
  const int i = (int)(tag & (unsigned long long)(K - 1));
  while (true) {
    unsigned long long o = *reinterpret_cast<volatile unsigned long long*>(&tab[i].owner);
    if (o == tag) return i;
    if (o == 0ull) {
      o = atomicCAS(&tab[i].owner, 0ull, tag);
      if (o == 0ull || o == tag) return i;
    }
    __nanosleep(256);   // held by a launch K ids older that is still running
  }
}

__device__ __forceinline__ int claim_launch_slot(LaunchSlot* tab) { return claim_slot<kLaunchSlots>(tab); }

// Called by the launch's last CTA (every CTA has finished with the slot):
// zero the counters, make that visible, then free the slot.
__device__ __forceinline__ void release_launch_slot(LaunchSlot* tab, int i) {
#pragma unroll
  for (int k = 0; k < 6; ++k) tab[i].c[k] = 0u;
  __threadfence();
  atomicExch(&tab[i].owner, 0ull);
}

}  // namespace lift
