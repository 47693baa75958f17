// Device-side dependency-counting task scheduler (CHOL_EXEC_SCHEDULER).
#pragma once
#include <cuda.h>
#include <cuda_runtime.h>

#include "../../include/chol.h"
#include "kernels.h"

namespace chol {
struct SchedState;
int sched_create(SchedState** out, int64_t N, int64_t nb, int bs, int sms, const chol_opts_t* opts, cudaStream_t s);
int sched_run(SchedState* st, const CUtensorMap& map, const StepParams& base, cudaStream_t s, int* nlaunch);
int sched_workers(const SchedState* st);
int sched_job_trace(const SchedState* st, uint64_t* out, int64_t cap, int64_t* njobs);
void sched_destroy(SchedState* st);
}  // namespace chol
