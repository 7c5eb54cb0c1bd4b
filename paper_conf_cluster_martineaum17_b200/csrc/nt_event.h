// nt_event.h -- event-based (Over Events, §V-B) variant of the tracker.
#pragma once
#include <cstdint>
#include <string>

#include "../../include/neutral_b200.h"
#include "nt_internal.h"

namespace nt {

struct EventState;
EventState* event_state_create();
void event_state_destroy(EventState* s);
void event_state_invalidate(EventState* s);   // particles re-injected: drop cached buffers
nt_status event_run_timestep(EventState* s, const TrackParams& tp, bool det, int sm_count,
                             cudaStream_t stream, uint32_t& launches, std::string& err);

}  // namespace nt
