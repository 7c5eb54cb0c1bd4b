// nt_event.cu -- event-based variant (placeholder until the queue kernels land).
#include "nt_event.h"

namespace nt {
struct EventState { int dummy; };
EventState* event_state_create() { return new EventState(); }
void event_state_destroy(EventState* s) { delete s; }
void event_state_invalidate(EventState*) {}
nt_status event_run_timestep(EventState*, const TrackParams&, bool, int, cudaStream_t,
                             uint32_t&, std::string& err) {
  err = "event mode not built yet";
  return NT_ERR_UNSUPPORTED;
}
}  // namespace nt
