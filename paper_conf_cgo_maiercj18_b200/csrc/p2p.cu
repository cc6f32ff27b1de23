// p2p.cu -- NEXT-4: flag signalling of the peer-memory halo
// exchange.  The halo rows themselves travel inside the step kernels (direct
// stores into the neighbours' band buffers, engine.cuh / hotspot_tb.cu); these
// two one-thread kernels order the launches of neighbouring bands:
//   step e  -> p2p_signal(e): fence.sc.sys, then st.release.sys of e into the
//              neighbours' flags;
//   p2p_wait(e): ld.acquire.sys polling of this band's own flags -> step e+1.
// A band starts launch e+1 only after both neighbours finished launch e: their
// halo stores for e have landed, and they no longer read the buffer parity
// that launch e+1 writes into them.
#include "p2p.cuh"

namespace kp {

__global__ void p2p_signal_kernel(unsigned* up_flag, unsigned* dn_flag, unsigned epoch) {
  asm volatile("fence.sc.sys;" ::: "memory");
  if (up_flag) asm volatile("st.release.sys.global.u32 [%0], %1;" ::"l"(up_flag), "r"(epoch) : "memory");
  if (dn_flag) asm volatile("st.release.sys.global.u32 [%0], %1;" ::"l"(dn_flag), "r"(epoch) : "memory");
}

__device__ __forceinline__ unsigned ld_acquire_sys(const unsigned* p) {
  unsigned v;
  asm volatile("ld.acquire.sys.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}

__global__ void p2p_wait_kernel(const unsigned* flags, int need_up, int need_dn, unsigned epoch) {
  unsigned polls = 0;
  for (;;) {
    const bool up = !need_up || (int)(ld_acquire_sys(flags) - epoch) >= 0;  // wrap-safe >=
    const bool dn = !need_dn || (int)(ld_acquire_sys(flags + 1) - epoch) >= 0;
    if (up && dn) break;
    if (++polls > (1u << 28)) __trap();  // a lost neighbour must not hang the GPU
    __nanosleep(64);
  }
}

cudaError_t p2p_signal(unsigned* up_flag, unsigned* dn_flag, unsigned epoch, cudaStream_t s) {
  p2p_signal_kernel<<<1, 1, 0, s>>>(up_flag, dn_flag, epoch);
  return cudaGetLastError();
}

cudaError_t p2p_wait(const unsigned* my_flags, int need_up, int need_dn, unsigned epoch, cudaStream_t s) {
  p2p_wait_kernel<<<1, 1, 0, s>>>(my_flags, need_up, need_dn, epoch);
  return cudaGetLastError();
}

}  // namespace kp
