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
// Track local particles [tp.lo, tp.hi) for one timestep with the event queues; adds the
// range's statistics into tp.stats_*.  Deterministic mode (det) writes flush records.
nt_status event_run_range(EventState* s, const TrackParams& tp, bool det, int sm_count,
                          cudaStream_t stream, uint32_t& launches, std::string& err);
// Iterations the device loop ran for the last range (synchronises the stream).
unsigned event_iterations(EventState* s, cudaStream_t stream);

}  // namespace nt
