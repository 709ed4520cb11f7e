/*
 * vsched.h — C ABI of libvsched: self-adaptive versioned tile tasks on B200.
 *
 * The calls follow the problem statement of Planas, Badia, Ayguade, Labarta,
 * "Self-Adaptive OmpSs Tasks in Heterogeneous Environments", IPDPS 2013
 * (PAPER.md line numbers L..., section in parentheses):
 *   - task functions with input/output/inout data (L231-242, Sec III)
 *   - several implementations of one task, "implements(main)"
 *     (L270-276, L298-351, Sec IV.A, Fig 4)
 *   - copy_deps data motion between address spaces (L220-230, L252-264)
 *   - taskwait / taskwait on / noflush (L243-246, L264-270)
 *   - scheduler plug-in and its options chosen by configuration (L277-288);
 *     lambda configurable (L438-440, footnote 4 L461)
 *   - versioning scheduler: TaskVersionSet <VersionId, ExecTime, #Exec> per
 *     DataSetSize group (L358-385, Table I), learning phase then earliest
 *     executor (L397-495, Fig 5)
 *   - statistics: Input/Output/Device Tx and per-version run counts (L515-536)
 * Readings where the paper is silent are numbered R1..R25 in DESIGN.md.
 *
 * Conventions
 *   - Every function returns vs_status (0 = VS_OK, negative = error) unless
 *     stated.  Synchronous misuse returns an error and sets vs_last_error().
 *   - Asynchronous failures (CUDA error, non-positive Cholesky pivot) are
 *     STICKY: they are returned by the next vs_wait_* call; afterwards only
 *     vs_stats*, vs_last_error and vs_destroy are valid.
 *   - Pointers passed as task data are NOT owned by the runtime.  The caller
 *     must not touch registered data between the submission of a task that
 *     uses it and the wait that covers it (OmpSs rule, L264-270).
 *   - "stream" arguments are cudaStream_t passed as void* (NULL = legacy
 *     default stream); no CUDA or torch type appears in this header.
 *   - Single submitting thread (OmpSs master-thread model, L213-215).
 */
#ifndef VSCHED_H
#define VSCHED_H

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif
#if defined(__GNUC__)
#pragma GCC visibility push(default)
#endif

typedef struct vs_runtime *vs_rt;
typedef int32_t vs_type_id;
typedef int32_t vs_version_id;
typedef int64_t vs_data_id;
typedef int64_t vs_task_id;

/* Access modes of a task parameter (StarSs clauses, L236-242). */
enum { VS_IN = 1, VS_OUT = 2, VS_INOUT = 3 };

typedef enum {
    VS_OK = 0,
    VS_E_INVAL = -1,     /* bad argument / unknown id */
    VS_E_NOMEM = -2,     /* host or device allocation failed */
    VS_E_CUDA = -3,      /* CUDA error (sticky when asynchronous) */
    VS_E_NOT_SPD = -4,   /* potrf found a non-positive pivot (sticky, R9) */
    VS_E_STATE = -5,     /* call not valid in the current state (e.g. after a sticky error) */
    VS_E_OVERLAP = -6,   /* registered regions partially overlap (R21) */
    VS_E_NODEV = -7,     /* no CUDA device / library built without a usable device */
    VS_E_IO = -8         /* timing-table file could not be read or written */
} vs_status;

/* Executors. */
enum { VS_EXEC_GPU = 0, /* tasks run on B200s */
       VS_EXEC_SIM = 1  /* no device: tasks take their durations from the timing
                           table on a virtual clock (DES); used for replay tests */ };
/* When a decision is taken (GPU executor). */
enum { VS_MODE_RUNAHEAD = 0, /* decide on the virtual clock as soon as predecessors are
                                decided; dependences are enforced on the device
                                ("look-ahead scheduling", L811) — default */
       VS_MODE_READY = 1     /* paper-literal: decide when predecessors have really
                                completed (L400-405) */ };
enum { VS_LEARN_HOLD = 0, VS_LEARN_RR = 1 };            /* reading R12 */
enum { VS_POLICY_VERSIONING = 0, VS_POLICY_FIXED = 1 };  /* FIXED = always fixed_version */
enum { VS_F32 = 0, VS_F64 = 1 };

/* Built-in tile task types (reading R5).  Tiles are b x b,
 * row-major, contiguous (leading dimension b), D6.  Parameters in order:
 *   VS_T_MATMUL : in A, in B, inout C        C += A * B            (Fig 1)
 *   VS_T_POTRF  : inout A                    A  = L, L*L^T = A     (lower, in place; L697-699)
 *   VS_T_TRSM   : in L, inout B              B  = B * L^{-T}       (right, lower, trans, non-unit)
 *   VS_T_SYRK   : in A, inout C              C -= A * A^T          (lower triangle only)
 *   VS_T_GEMM_NT: in A, in B, inout C        C -= A * B^T
 * The strict upper triangle of POTRF/SYRK tiles is neither read nor written (R7). */
enum { VS_T_MATMUL = 0, VS_T_POTRF = 1, VS_T_TRSM = 2, VS_T_SYRK = 3, VS_T_GEMM_NT = 4,
       VS_NUM_BUILTIN_TYPES = 5 };

/* Built-in versions (hand-written sm_100a kernels; "implements(main)" siblings). */
enum {
    VS_V_SIMT_F32 = 0,    /* IEEE fp32 FMA, fixed ascending-k order, smem staging + warp shuffles */
    VS_V_TC_3XTF32 = 1,   /* tcgen05/TMEM 3xTF32 (big*big + big*small + small*big) */
    VS_V_F64IN_F32IO = 2, /* fp32 in/out, fp64 arithmetic (DMMA), one rounding on store */
    VS_V_DFMA_F64 = 3,    /* fp64 tiles, SIMT DFMA */
    VS_V_DMMA_F64 = 4,    /* fp64 tiles, mma.sync f64 tensor cores */
    VS_V_TC_3XF16 = 5,    /* fp32 tiles, tcgen05 kind::f16 on row-scaled fp16 big/small halves of the
                             operands (reading R30); MATMUL, GEMM_NT, SYRK, and TRSM as X = B inv(L)^T
                             (R31); no POTRF.  Its in-operands
                             are read through a per-GPU cached "split form" that the runtime builds
                             (one conversion kernel per datum version, like a tile move) */
    VS_V_OZ_I8_F64 = 6,   /* fp64 tiles, tcgen05 kind::i8 Ozaki scheme (NEXT-4): each operand row as
                             7 int8 slices under a power-of-two row scale (a cached "slice form",
                             like tc_3xf16's split form), the 28 slice products with i + j <= 8
                             accumulated exactly in int32 TMEM (one accumulator per diagonal),
                             combined in fp64; MATMUL, GEMM_NT, SYRK; TRSM as X = B inv(L)^T
                             with the slice form of inv(L) (like tc_3xf16's R31); POTRF
                             recursive (DFMA diagonal blocks, DMMA panel trsm, Ozaki trailing
                             updates on slice forms built inside the task) */
    VS_NUM_BUILTIN_VERSIONS = 7
};

typedef struct {
    int exec;          /* VS_EXEC_GPU | VS_EXEC_SIM */
    int n_gpus;        /* number of devices driven by this runtime (workers' gpus 0..n_gpus-1) */
    int device_base;   /* CUDA ordinal of runtime gpu 0 (one process per GPU: LOCAL_RANK) */
    int slots_per_gpu; /* S workers (streams) per GPU (R16); S=1 is paper-literal */
    int lambda;        /* learning runs per version (L438-440, L461); default 3 (R10) */
    int policy;        /* VS_POLICY_VERSIONING | VS_POLICY_FIXED */
    int fixed_version; /* version index used by VS_POLICY_FIXED (a per-type index, see
                          vs_register_builtins); vs_submit returns VS_E_INVAL for a type that
                          has no runnable version of that index */
    int learning;      /* VS_LEARN_HOLD | VS_LEARN_RR */
    int mode;          /* VS_MODE_RUNAHEAD | VS_MODE_READY */
    int replay;        /* 1: the scheduler takes run times from the timing table, not from
                          measurements (bit-exact decisions, P8).  Implied by VS_EXEC_SIM. */
    int flush;         /* 1 (default): vs_wait_all copies written data back to its home
                          (OmpSs flush, L264-270) */
    int lookahead;     /* run-ahead window: at most this many issued-but-unfinished tasks
                          per GPU (0 = unlimited).  Keeps worker queues short so a task on
                          the critical path is not queued behind far-ahead work. */
    int priority;      /* 0: ready tasks in submission order (R15, paper-literal);
                          1: critical-path first (NEXT-4): ready order POTRF < TRSM < SYRK <
                          GEMM_NT < MATMUL < user types, and POTRF/TRSM/SYRK launched on a
                          high-priority stream of their worker (L711-718: potrf must run as
                          soon as it is ready);
                          2: bottom level first (NEXT-4, generic): ready order by the
                          longest path (in tasks) from the task to the end of the submitted
                          DAG, larger first, ties by id; same high-priority streams as 1 */
    int group_ratio_permille; /* 0: DataSetSize groups match exactly (R20).  r > 0: a new size
                          joins the first group of its type (creation order) within a factor
                          1 + r/1000 (range groups, future work L984-993; NEXT-3) */
    int ewma_weight;   /* 0: ExecTime is the arithmetic mean (L408-411).  w in 1..1024: recency-
                          weighted mean m += (x - m) * w / 1024 (footnote 3, L458-460; NEXT-3) */
    int locality_gbps; /* 0: earliest executor ignores data placement (paper).  g > 0: add
                          (bytes of the task not yet on the worker's GPU) / g GB/s to EFT
                          (locality-aware versioning, future work L978-984; NEXT-1) */
    int queue_depth;   /* 0: a ready task is assigned at once to its earliest executor,
                          whatever that worker's queue holds (paper, L414-422).  d > 0
                          (run-ahead, SIM): a ready task is assigned only while some worker
                          holds fewer than d virtual tasks (running + queued), and only to such
                          workers; (ready mode): fewer than d x group_tasks issued, unfinished
                          tasks.  The rest wait in the (priority) ready queue, so a task
                          released later on the critical path overtakes them (NEXT-4) */
    int group_tasks;   /* grouped launches (this build): up to this many consecutive tasks of
                          one worker whose version can share a launch (tc_3xf16 MATMUL /
                          GEMM_NT / SYRK) are enqueued as ONE kernel launch on the worker's
                          stream (no dependences inside a group: a task whose predecessor is
                          still pending flushes it first).  0 or 1: one launch per task */
    int group_wait_us; /* a pending group is launched after this many microseconds of host
                          time even if not full (and whenever the runtime has nothing else to
                          do, unless group_hold); 0 = default 20 */
    int group_hold;    /* 1: when the runtime has nothing else to do it launches only the
                          pending groups whose stream has no launched, unfinished kernel (the
                          stream would otherwise idle); the others keep collecting tasks until
                          group_wait_us.  Fewer, larger launches: the host issues ~1 launch per
                          2.5 tasks instead of ~1 per task in ready mode.  0: launch them all */
    int device_release; /* 1: device dependence tracker (a3; L400-405): ready mode, one GPU, one
                          process — at the start of a batch the runtime copies every task's
                          in-degree and CSR successor list to the GPU; the last CTA of a task's
                          last kernel (or a one-warp kernel after a user version) decrements
                          its successors' in-degrees and appends those reaching zero to a
                          host-mapped ready ring, which the host reads instead of counting
                          predecessors.  0: the host releases successors.  VS_TRACKER=device /
                          host overrides */
    const char *trace_path; /* non-NULL: every vs_wait_* (and vs_decision_log_clear) appends the
                          decision-log records completed since the previous append to this file
                          as JSON lines {"task", "type", "version", "worker", "phase",
                          "t_decide_ns", "t_start_ns", "t_end_ns"}; the string is copied */
    /* Device memory for tile replicas and operand forms (slabs of >= 1 GiB, or the request
     * size when that fails) comes from dev_alloc(cuda_device, bytes, alloc_user) when set
     * (e.g. a framework's caching allocator; NULL = out of memory) and is returned with
     * dev_free(cuda_device, ptr, alloc_user) at vs_destroy (dev_alloc without dev_free: never
     * returned).  NULL: cudaMalloc / cudaFree.  Control structures of the runtime (execution
     * records, rings, completion words) always use the CUDA allocator. */
    void *(*dev_alloc)(int device, size_t bytes, void *user);
    void (*dev_free)(int device, void *ptr, void *user);
    void *alloc_user;
    int stage;         /* n > 0 (default 32): transfer-ordered drive (reading R39; L515-532) — when a
                          fresh batch in ready mode with priority 2 on one GPU of one process reads
                          data homed in host memory, a list schedule of the batch fixes the order
                          in which those inputs cross the host link (critical path first, then
                          fewest unplanned input bytes, then the datum closest to its final
                          version, then weighted bottom level); the runtime copies them in that
                          order with at most n copies in flight, uses the planned position as the
                          ready order, and decides a task only once its inputs have arrived.
                          0: inputs move on demand when their reader is issued.  VS_STAGE=n
                          overrides */
} vs_config;

/* Fill *cfg with defaults: GPU, 1 gpu, base 0, 4 slots, lambda 3, versioning, hold,
 * run-ahead, live timing, flush.  Environment overrides applied by vs_create (L277-288):
 * VS_LAMBDA, VS_SLOTS, VS_POLICY(=versioning|fixed:<v>), VS_LEARNING(=hold|rr),
 * VS_MODE(=runahead|ready), VS_LOOKAHEAD(=n), VS_PRIORITY(=0|1|2), VS_QDEPTH(=d), VS_GROUP_HOLD(=0|1),
 * VS_GROUP(=tasks per grouped launch), VS_GROUP_US, VS_STAGE(=n).  Runtime options outside vs_config:
 * VS_TRACKER(=events|memops) dependence tracker on one GPU, VS_GROUP_DIST(=0|1, default 1)
 * grouped launches in a multi-rank job, VS_PREFETCH(=n, default 0) input-prefetch window on one
 * GPU, VS_TCF_PAIR(=0|1, default 0) CTA-pair variant of the tc_3xf16 GEMM. */
void vs_config_default(vs_config *cfg);

/* Create a runtime.  *out receives an opaque handle owning scheduler state, DAG,
 * data directory, CUDA streams/events and device replicas.
 * Errors: VS_E_INVAL (bad cfg), VS_E_NODEV (exec GPU but no device), VS_E_CUDA. */
int vs_create(const vs_config *cfg, vs_rt *out);
/* Wait for all tasks (no flush), release every resource.  Safe after a sticky error. */
int vs_destroy(vs_rt rt);
/* Last error message of this runtime (static storage until the next call); never NULL. */
const char *vs_last_error(vs_rt rt);

/* ---------------------------------------------------------- registration (a1) */
/* Declare a task type ("main implementation", L298-351) with nparams parameters
 * whose access modes are modes[i] in {VS_IN, VS_OUT, VS_INOUT}. */
int vs_type_create(vs_rt rt, const char *name, int nparams, const int *modes, vs_type_id *out);

/* A version launch function: enqueue the version's work for one task on `stream`
 * (a cudaStream_t).  dev_ptrs[i] is parameter i on the executing GPU, bytes[i] its
 * size.  Must not synchronise the stream, must touch only its parameters, must be
 * deterministic.  Return 0 on success. */
typedef int (*vs_launch_fn)(void *const *dev_ptrs, const int64_t *bytes, int nargs,
                            const void *scalars, size_t nscalar, void *stream, void *user);

/* Add a version to a type ("implements(main)", Fig 4).  All versions share the
 * type's parameters and modes (L306-308).  gpu_mask bit g = runnable on runtime gpu g
 * (the device clause, L339-345); a mask naming no configured gpu is VS_E_INVAL.
 * *out = version index within the type (0,1,...).  Versions must be added before the first
 * submission (VS_E_STATE after it).  The runtime times a user version with a CUDA event pair
 * around fn on the worker's stream (R17). */
int vs_version_add(vs_rt rt, vs_type_id type, const char *name, uint32_t gpu_mask,
                   vs_launch_fn fn, void *user, vs_version_id *out);

/* Register the five built-in tile task types for dtype, keeping the versions whose bit is
 * set in version_mask (bit = VS_V_*).  Versions each type actually gets:
 *   VS_F32: SIMT_F32, TC_3XTF32, F64IN_F32IO for all five types; TC_3XF16 for MATMUL,
 *           GEMM_NT, SYRK and TRSM (by inverse, R31) — not POTRF.
 *   VS_F64: DFMA_F64, DMMA_F64 and OZ_I8_F64 for all five types (OZ_I8_F64: TRSM by inverse,
 *           POTRF recursive with Ozaki-scheme trailing updates).
 * out_types[VS_T_*] receives the type ids.  Version INDICES are per type: inside each type
 * the kept versions are numbered 0, 1, ... in increasing VS_V_* order, skipping those the type
 * does not get, so the same index may name different versions in different types (e.g. with
 * every f32 version selected, index 3 is TC_3XF16 for MATMUL but does not exist for POTRF);
 * vs_version_name() maps an index back to its name.  Runnable on every gpu.
 * Errors: VS_E_INVAL if no version of dtype is selected. */
int vs_register_builtins(vs_rt rt, int dtype, uint32_t version_mask,
                         vs_type_id out_types[VS_NUM_BUILTIN_TYPES]);

/* ------------------------------------------------------------ data (a2, a8) */
/* Register a datum (a tile) living at ptr in the memory of `device` (-1 = host,
 * preferably pinned; g >= 0 = runtime gpu g).  Identical (ptr, bytes) returns the
 * same id; a partial overlap with a registered region is VS_E_OVERLAP (R21). */
int vs_data_register(vs_rt rt, void *ptr, int device, int64_t bytes, vs_data_id *out);

/* The caller modified datum d at its home outside any task (after a wait): every other
 * copy (device replica, cached remote copy, derived operand form) is stale and will be
 * re-fetched / rebuilt on next use.  Callers MUST call it after such a modification.
 * VS_E_STATE if a task writing d is still in flight. */
int vs_data_invalidate(vs_rt rt, vs_data_id d);

/* (Both invalidation calls first wait for copies back to the host that are still in flight.)
 * vs_data_invalidate of ids[0..n-1] (one call for a whole matrix of tiles); stops at, and
 * returns the error of, the first failing id. */
int vs_data_invalidate_n(vs_rt rt, const vs_data_id *ids, int64_t n);

/* ------------------------------------------------------------- submission (a2) */
/* Create a task instance: RAW/WAR/WAW edges on whole data (L236-242).  scalars
 * (may be NULL) are copied and passed to the version.  Execution happens inside
 * the vs_wait_* calls (the submitting thread joins the runtime, as at taskwait). */
int vs_submit(vs_rt rt, vs_type_id type, const vs_data_id *args, int nargs,
              const void *scalars, size_t nscalar, vs_task_id *out);

/* ----------------------------------------------------------- waits (a15) */
/* Every wait (and vs_create / vs_destroy) leaves the calling thread's current CUDA device
 * as it found it. */
int vs_wait_all(vs_rt rt);          /* taskwait: all tasks, then flush to home */
int vs_wait_all_noflush(vs_rt rt);  /* taskwait noflush (L267-270): all tasks; written data
                                       stay on the devices (copies back to the host that the
                                       runtime had already started are completed first) */
int vs_wait_on(vs_rt rt, vs_data_id d); /* taskwait on(d): d's last writer done; d valid at home */

/* ---------------------------------------------------------------- statistics */
typedef struct {
    int64_t tasks_submitted, tasks_completed, decisions;
    int64_t input_tx_bytes;   /* host -> any GPU, counted per destination (L529-532, R25) */
    int64_t output_tx_bytes;  /* any GPU -> host (L527-528) */
    int64_t device_tx_bytes;  /* GPU <-> GPU (L524-525) */
    int64_t n_groups;
    int64_t error_task;       /* task of the first sticky error, -1 if none */
    int64_t error_info;       /* potrf info (1-based pivot within the tile), or CUDA error code */
    int64_t host_ns_decide;   /* host time spent in decisions (scheduler overhead) */
    int64_t host_ns_issue;    /* host time spent issuing GPU work */
    int64_t virtual_now_ns;   /* DES clock */
    int64_t kernel_launches;  /* process-wide count of libvsched kernel launches */
    int64_t tracker;          /* dependence tracker in use: 1 = device completion words
                                 (stream memory operations), 0 = CUDA events */
    int64_t forms_built;      /* derived operand forms built (VS_V_TC_3XF16 split halves) */
    int64_t host_ns_poll;     /* host time polling device completions */
    int64_t host_ns_launch;   /* part of host_ns_issue spent enqueuing the version's kernels */
    int64_t host_ns_deps;     /* part of host_ns_issue spent enqueuing dependence waits / forms */
    int64_t host_loops;       /* iterations of the runtime's drive loop */
    int64_t host_ns_vevent;   /* host time advancing the virtual clock (run-ahead DES) */
    int64_t host_ns_flush;    /* host time launching pending grouped launches from the loop */
    int64_t host_idle_loops;  /* drive-loop iterations that found nothing to do */
    int64_t device_released;  /* tasks made ready by the device dependence tracker (a3) */
    int64_t host_ns_group_launch; /* host time inside grouped kernel launches */
    int64_t group_launches;   /* grouped kernel launches issued */
    int64_t gated_tasks;      /* ready tasks that waited for their host inputs to arrive before
                                 being decided (transfer-ordered drive, vs_config.stage) */
    int64_t host_ns_drive_setup; /* host time from entering a wait's drive to its first
                                 decisions issued (dependence tracker upload, bottom levels,
                                 transfer plan) */
    int64_t host_ns_poll_idle;   /* part of host_ns_poll spent in polls that found no completed
                                 task (the host waiting on the GPU) */
} vs_stats_t;
int vs_stats(vs_rt rt, vs_stats_t *out);

#define VS_MAX_VERSIONS 8
typedef struct {
    vs_type_id type;
    int64_t dataset_bytes;             /* DataSetSize (footnote 2) */
    int nversions;
    int reliable;                      /* 1 once every runnable version ran lambda times */
    int64_t first_reliable_decision;   /* 1-based decision index within the group, -1 if none */
    int64_t decisions;
    int64_t n[VS_MAX_VERSIONS];        /* #Exec (completed, measured) */
    int64_t mean_ns[VS_MAX_VERSIONS];  /* ExecTime = floor(sum/n) (R18), 0 if n = 0 */
    int64_t assigned[VS_MAX_VERSIONS]; /* decisions that picked this version */
} vs_group_stat_t;
int vs_group_count(vs_rt rt);
int vs_group_stat(vs_rt rt, int group_index, vs_group_stat_t *out);
/* Name of a type / of version v of a type (static storage owned by rt); NULL if invalid. */
const char *vs_type_name(vs_rt rt, vs_type_id t);
const char *vs_version_name(vs_rt rt, vs_type_id t, vs_version_id v);

/* Decision log: one record per decision, in decision order. */
typedef struct {
    vs_task_id task;
    int32_t version, worker;   /* worker = gpu * slots_per_gpu + slot */
    int32_t phase;             /* 0 learning, 1 reliable */
    vs_type_id type;           /* task type */
    int64_t t_decide_ns;       /* virtual (run-ahead / sim) or host clock (ready) */
    int64_t t_start_ns, t_end_ns; /* sim: virtual clock; gpu: GPU timeline of the version's
                                     start/end events (ns since runtime creation) */
    int64_t launch;               /* gpu: number of the kernel launch that ran a built-in
                                     version's task (tasks of one grouped launch share it;
                                     multi-kernel versions: the first), -1 otherwise */
} vs_decision_t;
/* Host wall-clock time at which each decision-log entry's task was enqueued on its
 * stream, on the t_start_ns timeline (system clock minus the same origin: the GPU's
 * %globaltimer follows the host's system clock); 0 if not issued (sim).  Same indexing
 * and (cap, n) protocol as vs_decision_log.  Diagnostic. */
int vs_decision_issue_ns(vs_rt rt, int64_t *out, int64_t cap, int64_t *n);
/* Copy up to cap records (from the beginning) into out; *n = total records. */
int vs_decision_log(vs_rt rt, vs_decision_t *out, int64_t cap, int64_t *n);
/* FNV-1a 64 over (task, version, worker, t_decide) of every record, little-endian int64
 * (identical definition in oracle/sched_model.py). */
uint64_t vs_decision_log_hash(vs_rt rt);
int vs_decision_log_clear(vs_rt rt);

/* ---------------------------------------------------- timing table (NEXT-2) */
/* Text format, one line per (type, group, version):
 *   <type name> <dataset bytes> <version name> <mean ns> <n>
 * dump writes the current TaskVersionSets; load merges (sum = mean*n, assigned = n)
 * and switches loaded groups to reliable when every runnable version has n >= lambda. */
int vs_table_dump(vs_rt rt, const char *path);
int vs_table_load(vs_rt rt, const char *path);
/* Replay/sim duration of (type, dataset bytes, version); used when exec = SIM or
 * replay = 1.  A missing entry during replay is VS_E_STATE. */
int vs_replay_set(vs_rt rt, vs_type_id type, int64_t dataset_bytes, vs_version_id v, int64_t ns);

/* ---------------------------------------------- application drivers (Fig 1, R5) */
/* Tiled matmul driver of Fig 1 (L164-172): for i<m, j<n, k<l submit
 * MATMUL(A[i*l+k], B[k*n+j], C[i*n+j]).  A, B, C are arrays of data ids. */
int vs_app_matmul(vs_rt rt, vs_type_id matmul_type, int m, int l, int n,
                  const vs_data_id *A, const vs_data_id *B, const vs_data_id *C);
/* Right-looking lower tiled Cholesky (R5): A[i*nt+j] for i >= j, types[VS_T_*]. */
int vs_app_cholesky(vs_rt rt, const vs_type_id types[VS_NUM_BUILTIN_TYPES], int nt,
                    const vs_data_id *A);
/* Order the next drive (the device work of the next vs_wait_*) after a CUDA event the caller
 * recorded on its own stream (cudaEvent_t passed as void*; the caller keeps it alive until
 * that wait returns), e.g. the kernels that produced the batch's device-homed inputs: every
 * stream of the runtime waits for it on the device, so the runtime's host-side setup of the
 * drive (dependence tracker upload, bottom levels, transfer plan) overlaps the caller's work
 * instead of following a host synchronisation.  Consumed by that drive.  No-op in SIM. */
int vs_depend_on_event(vs_rt rt, void *cuda_event);
/* Transfer plan of the submitted batch before it starts (vs_config.stage, reading R39): the ids
 * of the host-homed data it reads, in the order a transfer-ordered drive copies them to the
 * GPU.  Writes min(cap, total) ids to out (caller-owned; may be NULL when cap = 0) and the
 * total to *n (0 when no task of the batch reads host-only data).  Starts nothing; any
 * executor.  VS_E_STATE once the batch has started (a wait has driven it). */
int vs_transfer_plan(vs_rt rt, vs_data_id *out, int64_t cap, int64_t *n);

/* ----------------------------------------------------- direct tile kernels */
/* Enqueue one built-in tile task version on `stream` on the current device, outside
 * the runtime (used by parity tests and the smoke check).  ptrs as in VS_T_* order,
 * device pointers, tiles b x b contiguous.  dinfo: device int32 receiving potrf's info
 * (may be NULL for other types).  Returns VS_E_INVAL for an unknown (type, version)
 * or an unsupported b (b must be a multiple of 64, 64 <= b <= 4096). */
int vs_tile_run(int type, int version, int b, void *const *ptrs, int *dinfo, void *stream);

/* Derived operand forms (reading R30).  vs_operand_form returns the form (0 = the tile
 * itself, 1 = row split form, 2 = column split form, i.e. the row split form of the
 * transposed tile, 3 = row split form of inv(L)) in which `version` reads parameter `param`
 * of built-in `type`;
 * vs_form_bytes the size of a form of a b x b tile (0 for form 0).
 * vs_form_make enqueues the conversion of the b x b tile `src` (fp32; fp64 for forms 4, 5) into `dst`
 * (vs_form_bytes bytes, device memory, 16-byte aligned) on `stream`.
 * vs_tile_run_prepared is vs_tile_run with the forms prepared by the caller (no
 * conversion): ptrs holds 2 * nparams pointers, ptrs[i] = the tile of parameter i (device),
 * ptrs[nparams + i] = its form (ignored for form 0) — the kernels the runtime launches for a
 * task.  Form 3 (TRSM of VS_V_TC_3XF16) = row split form of inv(L) for the lower triangle L
 * of the tile (reading R31).  Forms 4 / 5 / 6 (VS_V_OZ_I8_F64) = int8 slice form of the
 * rows (A role) / of the columns (matmul B) / of the rows in the B role of an NT product, of a
 * b x b fp64 tile; form 7 (TRSM of VS_V_OZ_I8_F64) = the B-role slice form of the rows of inv(L)
 * for the lower triangle L of a b x b fp64 tile.  VS_E_INVAL on bad arguments. */
int vs_operand_form(int type, int version, int param);
int64_t vs_form_bytes(int form, int b);
int vs_form_make(int form, int b, const void *src, void *dst, void *stream);
int vs_tile_run_prepared(int type, int version, int b, void *const *ptrs, int *dinfo, void *stream);

/* ---------------------------------------------------------- input generator */
/* Device counter-based generator, bit-identical to vsgen.uniform_idx:
 *   u(seed, idx) = (splitmix64((seed << 40) | idx) >> 40) * 2^-23 - 1.
 * Writes a rows x cols matrix (global index r*cols+c) as dtype VS_F32/VS_F64 into
 * dev_out: row-major if tile_b == 0, else tile-major (tiles tile_b x tile_b row-major,
 * tile (I,J) at offset (I*(cols/tile_b)+J)*tile_b^2). */
int vs_gen_uniform(uint64_t seed, int64_t rows, int64_t cols, int dtype, int tile_b,
                   void *dev_out, void *stream);
/* SPD recipe R8: S_rc = u(seed, max(r,c)*n + min(r,c)); diagonal fl(S_rr + alpha) with
 * alpha = 2.5*sqrt(n) (n >= 256) else n, computed in fp64.  Layout as vs_gen_uniform. */
int vs_gen_spd(uint64_t seed, int64_t n, int dtype, int tile_b, void *dev_out, void *stream);

/* One tile_b x tile_b tile at global tile coordinates (ti, tj) of the rows x cols uniform
 * matrix (spd = 0) or of the cols x cols SPD matrix (spd = 1), row-major, same values as
 * vs_gen_uniform / vs_gen_spd (used by ranks that own only some tiles). */
int vs_gen_tile(uint64_t seed, int64_t rows, int64_t cols, int dtype, int tile_b, int64_t ti, int64_t tj, int spd,
                void *dev_out, void *stream);

/* ------------------------------------------- one process per GPU */
/* Join a job of nranks processes on one node as `rank`.  Every rank submits the SAME task
 * graph; a task is executed only by the rank owning its written datum (owner computes,
 * vs_data_set_owner), and is retired at once elsewhere.  A rank reading a datum owned by
 * another rank copies it over NVLink from the owner's memory (a CUDA IPC pointer given at
 * registration) after the producing task's completion tag is visible: tags live in the
 * POSIX shared-memory segment shm_name (created by rank 0, which must call first; the
 * binding orders the calls with a barrier) registered with every rank's GPU, so the wait
 * is a stream memory operation on the device, with no host round trip.  Both decision modes
 * work (ready mode parks a task until its remote predecessors' tags are visible).
 * Restrictions: inside a graph a rank never overwrites a datum another rank may still be
 * copying (true of vs_app_matmul / vs_app_cholesky with owner computes); between graphs the
 * caller must not modify its owned data outside tasks (e.g. restore inputs) before every rank
 * has returned from its vs_wait_all of the previous graph (a barrier), and other ranks must
 * not read them before the modification is complete (a second barrier; see bench.py).  Must
 * precede submissions. */
int vs_dist_init(vs_rt rt, int rank, int nranks, const char *shm_name);
/* Datum d is owned by rank `owner` (its pointer is then the owner's memory, opened with
 * vs_ipc_open); data registered without this call belong to the calling rank. */
int vs_data_set_owner(vs_rt rt, vs_data_id d, int owner);
/* CUDA IPC without CUDA types: export a device pointer as a 64-byte handle + byte offset in
 * its allocation; open a peer handle (pointer valid in this process); close an opened base. */
int vs_ipc_export(const void *dev_ptr, unsigned char handle[64], uint64_t *offset);
int vs_ipc_open(const unsigned char handle[64], uint64_t offset, void **dev_ptr);
int vs_ipc_close(void *base_ptr);

/* CUDA ordinal of runtime gpu g (device_base + g), VS_E_INVAL if g is not a gpu of rt (SIM
 * runtimes have none).  One process per GPU: every rank's runtime drives its own device. */
int vs_gpu_ordinal(vs_rt rt, int g);

/* Library build information (never NULL). */
const char *vs_build_info(void);

#if defined(__GNUC__)
#pragma GCC visibility pop
#endif
#ifdef __cplusplus
}
#endif
#endif /* VSCHED_H */
