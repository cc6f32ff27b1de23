// p2p.cuh -- NEXT-4: epoch flags for the peer-memory halo exchange of the
// banded Hotspot (p2p.cu).  Each band owns two flags in device memory, written
// by its neighbours over NVLink (flag 0: "upper band finished launch e",
// flag 1: "lower band finished launch e").
#pragma once
#include <cuda_runtime.h>

namespace kp {

// after a step launch: make this band's halo stores visible system-wide, then
// publish `epoch` into the neighbours' flags (nullptr: no neighbour)
cudaError_t p2p_signal(unsigned* up_flag, unsigned* dn_flag, unsigned epoch, cudaStream_t s);
// before the next step launch: wait until each present neighbour has
// published >= epoch into this band's flags (watchdog: traps after ~2^28 polls)
cudaError_t p2p_wait(const unsigned* my_flags, int need_up, int need_dn, unsigned epoch, cudaStream_t s);

}  // namespace kp
