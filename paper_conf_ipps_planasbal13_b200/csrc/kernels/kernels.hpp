// kernels.hpp — internal interface between the runtime and the sm_100a tile kernels.
// Not part of the public ABI (see include/vsched.h).
#pragma once
#include <cuda_runtime.h>
#include <stdint.h>

#include <atomic>

namespace vsk {

// Process-wide count of kernels launched by libvsched (reported as gpu_launches).
inline std::atomic<long long> &launch_counter()
{
    static std::atomic<long long> c{0};
    return c;
}
inline void count_launch() { launch_counter().fetch_add(1, std::memory_order_relaxed); }
// Kernels a version launches for itself that carry no execution record (e.g. the operand
// forms oz_i8_f64's POTRF builds for its trailing updates): reported in the launch count, but
// not part of a task's kernel count (the completion of its record-carrying kernels).
inline std::atomic<long long> &aux_launch_counter()
{
    static std::atomic<long long> c{0};
    return c;
}
inline void count_launch_aux() { aux_launch_counter().fetch_add(1, std::memory_order_relaxed); }

// Device dependence tracker (a3): in-degrees and CSR successor lists of
// the tasks of one drive, in device memory of the runtime's GPU, built by the runtime at the
// start of the drive.  Task index = task id - first id of the batch.  The last CTA of a task's
// last kernel decrements the in-degree of each successor; a successor whose count reaches zero
// is appended to the host-mapped ready ring (entry = epoch << 32 | index + 1), which the host
// reads instead of counting predecessors itself.
struct DevTracker {
    int *indeg = nullptr;                    // [T] predecessors not yet complete
    const int *succ_off = nullptr;           // [T + 1]
    const int *succ = nullptr;               // [E]
    unsigned long long *rdy_ctr = nullptr;   // device counter of ready-ring entries
    unsigned long long *rdy_ring = nullptr;  // host-mapped ring (kRingCap entries, 0 = empty)
    unsigned long long epoch = 0;            // drive number (stale entries are ignored)
};

// Per-task execution record passed to every kernel of a built-in version (task_ctx.cuh).
// slot: device memory {start_min, end_max, ticket}; host: host-mapped {start, end,
// kernels completed, pad}.
// A default TaskCtx (nullptrs) disables recording (direct vs_tile_run calls).
struct TaskCtx {
    unsigned long long *slot = nullptr;   // device {~start min, end max, CTA ticket, CTA busy sum, longest CTA, -}
    unsigned long long *host = nullptr;   // host-mapped {~start, end, kernels done, exec time}
    unsigned int ncta = 0;   // CTAs of the task in the launch (0: the whole grid)
    unsigned int nsm = 0;    // SMs of the device
    unsigned int occ = 0;    // resident CTAs per SM of the kernel (occupancy; 0 = 1), set per launch
    // completion ring (host-mapped): the last CTA of every kernel of the task appends `tag`
    // at ring[atomicAdd(ring_ctr) % kRingCap], so the host reads completions in O(completed)
    unsigned long long *ring_ctr = nullptr;   // device counter of appended entries
    unsigned long long *ring = nullptr;       // host-mapped entries (0 = empty)
    unsigned long long tag = 0;               // task id + 1
    // device dependence release (a3): null = the host releases successors
    const DevTracker *trk = nullptr;
    int tidx = 0;              // task index in trk
    unsigned int nkern = 0;    // kernels of the task: the last one releases
};
constexpr unsigned long long kRingCap = 1ull << 16;

// Task types / versions use the VS_T_* / VS_V_* numbering of vsched.h.
// Returns 0 on success, -1 for an unsupported (type, version, b).
int launch_builtin(int type, int version, int b, void *const *p, int *dinfo, cudaStream_t s,
                   const TaskCtx &ctx = TaskCtx());
// Kernels launch_builtin enqueues for (type, version, b) (counted once by capturing a launch
// into a CUDA graph; cached), -1 if unsupported.
int builtin_kernel_count(int type, int version, int b);
// One-warp kernel doing only the dependence release of ctx (after a user version's work).
int launch_release(const TaskCtx &ctx, cudaStream_t s);
bool builtin_supported(int type, int version, int b);
// Element size in bytes for a version (4 for f32-io versions, 8 for f64).
int builtin_elem_bytes(int version);

// Operand forms: a version may read an in-parameter through a derived copy of the tile
// that the runtime builds and caches per (datum version, GPU), like a replica (a8).
// FORM_INV_L: row split form of inv(L) for the lower triangle L of a tile (TRSM by GEMM).
// Pointer layout of launch_builtin / group_add for versions with forms: p[i] = the tile
// of parameter i, p[nparams + i] = its form (nparams = builtin_nparams(type)).
// FORM_OZ_ROWS / FORM_OZ_COLS / FORM_OZ_ROWS_B: int8 slice forms of the rows (A role,
// 128-row groups) / columns (matmul B, 64-row groups) / rows (NT B role, 64-row groups) of
// an fp64 tile (oz_i8_f64, tc_oz.cuh).
// FORM_OZ_INV_L: int8 slice form (B role) of the rows of inv(L) for the lower triangle L of an
// fp64 tile (TRSM of oz_i8_f64 as X = B inv(L)^T, like tc_3xf16's FORM_INV_L).
enum { FORM_RAW = 0, FORM_SPLIT_ROWS = 1, FORM_SPLIT_COLS = 2, FORM_INV_L = 3, FORM_OZ_ROWS = 4, FORM_OZ_COLS = 5,
       FORM_OZ_ROWS_B = 6, FORM_OZ_INV_L = 7, NUM_FORMS = 8 };
inline bool form_is_f64(int f) { return f == FORM_OZ_ROWS || f == FORM_OZ_COLS || f == FORM_OZ_ROWS_B || f == FORM_OZ_INV_L; }
int builtin_nparams(int type);
int builtin_operand_form(int type, int version, int param);
size_t form_bytes(int form, int b);
// Build the form of the b x b fp32 tile src into dst (form_bytes) on stream s.
int make_form(int form, int b, const void *src, void *dst, cudaStream_t s);

// Grouped launches: versions whose tasks can share one kernel launch with other tasks of
// the same kind (tc_3xf16 MATMUL / GEMM_NT / SYRK: one grouped tcgen05 GEMM launch).
// group_kind() = 0 for versions that cannot be grouped.  A group is filled with
// group_add() (ptrs as for launch_builtin, ctx of the task; returns the task's CTA count,
// or -1 if it does not fit / is unsupported) and launched by group_launch().
struct TaskGroup;
int group_kind(int type, int version, int b);
TaskGroup *group_new();
void group_free(TaskGroup *g);
int group_size(const TaskGroup *g);
int group_ctas(const TaskGroup *g);
int group_add(TaskGroup *g, int type, int version, int b, void *const *p, const TaskCtx &ctx);
int group_launch(TaskGroup *g, cudaStream_t s);   // launches and empties the group

int gen_uniform(uint64_t seed, int64_t rows, int64_t cols, int dtype, int tile_b, void *out,
                cudaStream_t s);
int gen_spd(uint64_t seed, int64_t n, int dtype, int tile_b, void *out, cudaStream_t s);
int gen_tile(uint64_t seed, int64_t rows, int64_t cols, int dtype, int b, int64_t ti, int64_t tj, int spd, void *out,
             cudaStream_t s);

}  // namespace vsk
