// Host-side task graph of Algorithm 1 and its bottom levels (dag.cpp).
#pragma once
#include <cstdint>
#include <utility>
#include <vector>

namespace chol {
// edges (pred, succ) between dense task ids (taskid.h); type_of[id] = 0..3
void build_task_dag(int64_t N, std::vector<std::pair<int64_t, int64_t>>& edges, std::vector<int>& type_of);
// bottom level of every task (own weight w[type] included)
std::vector<double> bottom_levels(int64_t N, const double w[4]);
inline int tile_owner_h(int64_t i, int64_t j, int p, int q) { return (int)((i % p) * q + (j % q)); }
void dist_layout(int64_t N, int p, int q, int rank, std::vector<int>& slot_map, int* nowned, int* ncached);
void owner_slots(int64_t N, int p, int q, std::vector<int>& out);
}  // namespace chol
