"""paper_conf_ipps_planasbal13_b200 — Python binding of libvsched (include/vsched.h).

Argument marshalling only: every step of the hot path (scheduling decisions, dependence
tracking, data movement, tile kernels) runs inside libvsched.so (C++ / CUDA sm_100a).
The binding never falls back to Python or CPU code: if the library is missing it raises.

Names follow the C ABI (``vs_create``, ``vs_submit``, ...).  ``Runtime`` is a small
convenience holder that calls the same functions.
"""
from __future__ import annotations

import ctypes
import os
from ctypes import POINTER, Structure, c_char_p, c_double, c_int, c_int32, c_int64, c_size_t, c_uint32, c_uint64, c_void_p

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_HERE, "libvsched.so")

# ---- constants (mirror vsched.h) ----
VS_IN, VS_OUT, VS_INOUT = 1, 2, 3
VS_OK, VS_E_INVAL, VS_E_NOMEM, VS_E_CUDA, VS_E_NOT_SPD, VS_E_STATE, VS_E_OVERLAP, VS_E_NODEV, VS_E_IO = \
    0, -1, -2, -3, -4, -5, -6, -7, -8
VS_EXEC_GPU, VS_EXEC_SIM = 0, 1
VS_MODE_RUNAHEAD, VS_MODE_READY = 0, 1
VS_LEARN_HOLD, VS_LEARN_RR = 0, 1
VS_POLICY_VERSIONING, VS_POLICY_FIXED = 0, 1
VS_F32, VS_F64 = 0, 1
VS_T_MATMUL, VS_T_POTRF, VS_T_TRSM, VS_T_SYRK, VS_T_GEMM_NT = range(5)
VS_NUM_BUILTIN_TYPES = 5
VS_V_SIMT_F32, VS_V_TC_3XTF32, VS_V_F64IN_F32IO, VS_V_DFMA_F64, VS_V_DMMA_F64, VS_V_TC_3XF16, VS_V_OZ_I8_F64 = range(7)
VS_MAX_VERSIONS = 8
VERSION_NAMES = ["simt_f32", "tc_3xtf32", "f64in_f32io", "dfma_f64", "dmma_f64", "tc_3xf16", "oz_i8_f64"]
TYPE_NAMES = ["MATMUL", "POTRF", "TRSM", "SYRK", "GEMM_NT"]

ERRORS = {0: "VS_OK", -1: "VS_E_INVAL", -2: "VS_E_NOMEM", -3: "VS_E_CUDA", -4: "VS_E_NOT_SPD",
          -5: "VS_E_STATE", -6: "VS_E_OVERLAP", -7: "VS_E_NODEV", -8: "VS_E_IO"}


class vs_config(Structure):
    _fields_ = [("exec", c_int), ("n_gpus", c_int), ("device_base", c_int), ("slots_per_gpu", c_int),
                ("lambda_", c_int), ("policy", c_int), ("fixed_version", c_int), ("learning", c_int),
                ("mode", c_int), ("replay", c_int), ("flush", c_int), ("lookahead", c_int), ("priority", c_int),
                ("group_ratio_permille", c_int), ("ewma_weight", c_int), ("locality_gbps", c_int),
                ("queue_depth", c_int), ("group_tasks", c_int), ("group_wait_us", c_int), ("group_hold", c_int),
                ("device_release", c_int), ("trace_path", c_char_p), ("dev_alloc", c_void_p), ("dev_free", c_void_p),
                ("alloc_user", c_void_p), ("stage", c_int)]


# device allocator hooks of vs_config (dev_alloc / dev_free)
VS_DEV_ALLOC_FN = ctypes.CFUNCTYPE(c_void_p, c_int, c_size_t, c_void_p)
VS_DEV_FREE_FN = ctypes.CFUNCTYPE(None, c_int, c_void_p, c_void_p)


class vs_stats_t(Structure):
    _fields_ = [(n, c_int64) for n in (
        "tasks_submitted", "tasks_completed", "decisions", "input_tx_bytes", "output_tx_bytes", "device_tx_bytes",
        "n_groups", "error_task", "error_info", "host_ns_decide", "host_ns_issue", "virtual_now_ns",
        "kernel_launches", "tracker", "forms_built", "host_ns_poll", "host_ns_launch", "host_ns_deps", "host_loops", "host_ns_vevent", "host_ns_flush",
        "host_idle_loops", "device_released", "host_ns_group_launch", "group_launches", "gated_tasks", "host_ns_drive_setup", "host_ns_poll_idle")]


class vs_group_stat_t(Structure):
    _fields_ = [("type", c_int32), ("dataset_bytes", c_int64), ("nversions", c_int), ("reliable", c_int),
                ("first_reliable_decision", c_int64), ("decisions", c_int64),
                ("n", c_int64 * VS_MAX_VERSIONS), ("mean_ns", c_int64 * VS_MAX_VERSIONS),
                ("assigned", c_int64 * VS_MAX_VERSIONS)]


class vs_decision_t(Structure):
    _fields_ = [("task", c_int64), ("version", c_int32), ("worker", c_int32), ("phase", c_int32), ("type", c_int32),
                ("t_decide_ns", c_int64), ("t_start_ns", c_int64), ("t_end_ns", c_int64), ("launch", c_int64)]


VS_LAUNCH_FN = ctypes.CFUNCTYPE(c_int, POINTER(c_void_p), POINTER(c_int64), c_int, c_void_p, c_size_t, c_void_p,
                                c_void_p)

_lib = None


class VSError(RuntimeError):
    def __init__(self, code, msg=""):
        super().__init__("%s (%d): %s" % (ERRORS.get(code, "?"), code, msg))
        self.code = code


def lib():
    """Load libvsched.so (in-tree build).  Raises if it is missing: there is no fallback."""
    global _lib
    if _lib is not None:
        return _lib
    if not os.path.exists(LIB_PATH):
        raise ImportError("libvsched.so not built (run python -c 'import __graft_entry__ as g; g.build()')")
    L = ctypes.CDLL(LIB_PATH)
    rt = c_void_p
    sig = {
        "vs_config_default": (None, [POINTER(vs_config)]),
        "vs_create": (c_int, [POINTER(vs_config), POINTER(rt)]),
        "vs_destroy": (c_int, [rt]),
        "vs_last_error": (c_char_p, [rt]),
        "vs_type_create": (c_int, [rt, c_char_p, c_int, POINTER(c_int), POINTER(c_int32)]),
        "vs_version_add": (c_int, [rt, c_int32, c_char_p, c_uint32, VS_LAUNCH_FN, c_void_p, POINTER(c_int32)]),
        "vs_register_builtins": (c_int, [rt, c_int, c_uint32, POINTER(c_int32)]),
        "vs_data_register": (c_int, [rt, c_void_p, c_int, c_int64, POINTER(c_int64)]),
        "vs_submit": (c_int, [rt, c_int32, POINTER(c_int64), c_int, c_void_p, c_size_t, POINTER(c_int64)]),
        "vs_wait_all": (c_int, [rt]),
        "vs_wait_all_noflush": (c_int, [rt]),
        "vs_wait_on": (c_int, [rt, c_int64]),
        "vs_stats": (c_int, [rt, POINTER(vs_stats_t)]),
        "vs_group_count": (c_int, [rt]),
        "vs_group_stat": (c_int, [rt, c_int, POINTER(vs_group_stat_t)]),
        "vs_type_name": (c_char_p, [rt, c_int32]),
        "vs_version_name": (c_char_p, [rt, c_int32, c_int32]),
        "vs_decision_log": (c_int, [rt, POINTER(vs_decision_t), c_int64, POINTER(c_int64)]),
        "vs_decision_log_hash": (c_uint64, [rt]),
        "vs_decision_log_clear": (c_int, [rt]),
        "vs_table_dump": (c_int, [rt, c_char_p]),
        "vs_table_load": (c_int, [rt, c_char_p]),
        "vs_replay_set": (c_int, [rt, c_int32, c_int64, c_int32, c_int64]),
        "vs_app_matmul": (c_int, [rt, c_int32, c_int, c_int, c_int, POINTER(c_int64), POINTER(c_int64),
                                  POINTER(c_int64)]),
        "vs_app_cholesky": (c_int, [rt, POINTER(c_int32), c_int, POINTER(c_int64)]),
        "vs_transfer_plan": (c_int, [rt, POINTER(c_int64), c_int64, POINTER(c_int64)]),
        "vs_depend_on_event": (c_int, [rt, c_void_p]),
        "vs_tile_run": (c_int, [c_int, c_int, c_int, POINTER(c_void_p), c_void_p, c_void_p]),
        "vs_gen_uniform": (c_int, [c_uint64, c_int64, c_int64, c_int, c_int, c_void_p, c_void_p]),
        "vs_gen_spd": (c_int, [c_uint64, c_int64, c_int, c_int, c_void_p, c_void_p]),
        "vs_build_info": (c_char_p, []),
        "vs_gen_tile": (c_int, [c_uint64, c_int64, c_int64, c_int, c_int, c_int64, c_int64, c_int, c_void_p, c_void_p]),
        "vs_dist_init": (c_int, [rt, c_int, c_int, c_char_p]),
        "vs_data_set_owner": (c_int, [rt, c_int64, c_int]),
        "vs_ipc_export": (c_int, [c_void_p, ctypes.c_char * 64, POINTER(c_uint64)]),
        "vs_ipc_open": (c_int, [ctypes.c_char * 64, c_uint64, POINTER(c_void_p)]),
        "vs_ipc_close": (c_int, [c_void_p]),
        "vs_data_invalidate": (c_int, [rt, c_int64]),
        "vs_data_invalidate_n": (c_int, [rt, c_void_p, c_int64]),
        "vs_operand_form": (c_int, [c_int, c_int, c_int]),
        "vs_form_bytes": (c_int64, [c_int, c_int]),
        "vs_form_make": (c_int, [c_int, c_int, c_void_p, c_void_p, c_void_p]),
        "vs_tile_run_prepared": (c_int, [c_int, c_int, c_int, POINTER(c_void_p), c_void_p, c_void_p]),
        "vs_decision_issue_ns": (c_int, [rt, POINTER(c_int64), c_int64, POINTER(c_int64)]),
        "vs_gpu_ordinal": (c_int, [rt, c_int]),
    }
    for name, (res, args) in sig.items():
        f = getattr(L, name)
        f.restype = res
        f.argtypes = args
    _lib = L
    return L


EXPORTED = ["vs_config_default", "vs_create", "vs_destroy", "vs_last_error", "vs_type_create", "vs_version_add",
            "vs_register_builtins", "vs_data_register", "vs_submit", "vs_wait_all", "vs_wait_all_noflush",
            "vs_wait_on", "vs_stats", "vs_group_count", "vs_group_stat", "vs_type_name", "vs_version_name",
            "vs_decision_log", "vs_decision_log_hash", "vs_decision_log_clear", "vs_table_dump", "vs_table_load",
            "vs_replay_set", "vs_app_matmul", "vs_app_cholesky", "vs_transfer_plan", "vs_depend_on_event", "vs_tile_run", "vs_gen_uniform", "vs_gen_spd",
            "vs_build_info", "vs_gen_tile", "vs_dist_init", "vs_data_set_owner", "vs_ipc_export", "vs_ipc_open",
            "vs_ipc_close", "vs_data_invalidate", "vs_data_invalidate_n", "vs_operand_form", "vs_form_bytes", "vs_form_make",
            "vs_tile_run_prepared", "vs_decision_issue_ns", "vs_gpu_ordinal"]


def _ids(seq, ctype=c_int64):
    arr = (ctype * len(seq))(*seq)
    return arr


# ------------------------------------------------------------------ thin wrappers
def vs_config_default(**kw) -> vs_config:
    """vs_config with defaults, keyword overrides on top.  trace_path: str; dev_alloc /
    dev_free: ctypes callbacks (VS_DEV_ALLOC_FN / VS_DEV_FREE_FN) kept alive by the config."""
    c = vs_config()
    lib().vs_config_default(ctypes.byref(c))
    c._keep = []
    for k, v in kw.items():
        if k == "trace_path" and isinstance(v, str):
            v = v.encode()
            c._keep.append(v)
        elif k in ("dev_alloc", "dev_free") and v is not None and not isinstance(v, int):
            c._keep.append(v)
            v = ctypes.cast(v, c_void_p).value
        setattr(c, "lambda_" if k == "lam" else k, v)
    return c


def vs_tile_run(ttype, version, b, ptrs, dinfo=0, stream=0):
    """Enqueue one built-in tile task version (device pointers as ints)."""
    arr = (c_void_p * len(ptrs))(*ptrs)
    r = lib().vs_tile_run(ttype, version, b, arr, c_void_p(dinfo or None), c_void_p(stream or None))
    if r:
        raise VSError(r, "vs_tile_run(type=%d, version=%d, b=%d)" % (ttype, version, b))


def vs_operand_form(ttype, version, param):
    return lib().vs_operand_form(ttype, version, param)


def vs_form_bytes(form, b):
    return lib().vs_form_bytes(form, b)


def vs_form_make(form, b, src_ptr, dst_ptr, stream=0):
    r = lib().vs_form_make(form, b, c_void_p(src_ptr), c_void_p(dst_ptr), c_void_p(stream or None))
    if r:
        raise VSError(r, "vs_form_make(form=%d, b=%d)" % (form, b))


def vs_tile_run_prepared(ttype, version, b, ptrs, dinfo=0, stream=0):
    """vs_tile_run with the operands already in the version's forms (vs_operand_form)."""
    arr = (c_void_p * len(ptrs))(*ptrs)
    r = lib().vs_tile_run_prepared(ttype, version, b, arr, c_void_p(dinfo or None), c_void_p(stream or None))
    if r:
        raise VSError(r, "vs_tile_run_prepared(type=%d, version=%d, b=%d)" % (ttype, version, b))


def vs_gen_uniform(seed, rows, cols, dtype, tile_b, dev_ptr, stream=0):
    r = lib().vs_gen_uniform(seed, rows, cols, dtype, tile_b, c_void_p(dev_ptr), c_void_p(stream or None))
    if r:
        raise VSError(r, "vs_gen_uniform")


def vs_gen_spd(seed, n, dtype, tile_b, dev_ptr, stream=0):
    r = lib().vs_gen_spd(seed, n, dtype, tile_b, c_void_p(dev_ptr), c_void_p(stream or None))
    if r:
        raise VSError(r, "vs_gen_spd")


def vs_build_info() -> str:
    return lib().vs_build_info().decode()


def vs_gen_tile(seed, rows, cols, dtype, tile_b, ti, tj, spd, dev_ptr, stream=0):
    r = lib().vs_gen_tile(seed, rows, cols, dtype, tile_b, ti, tj, spd, c_void_p(dev_ptr), c_void_p(stream or None))
    if r:
        raise VSError(r, "vs_gen_tile")


def vs_ipc_export(dev_ptr):
    """-> (64-byte handle as bytes, offset) of a device pointer."""
    h = (ctypes.c_char * 64)()
    off = c_uint64()
    r = lib().vs_ipc_export(c_void_p(dev_ptr), h, ctypes.byref(off))
    if r:
        raise VSError(r, "vs_ipc_export")
    return bytes(h.raw), off.value


def vs_ipc_open(handle: bytes, offset: int) -> int:
    h = (ctypes.c_char * 64).from_buffer_copy(handle)
    p = c_void_p()
    r = lib().vs_ipc_open(h, offset, ctypes.byref(p))
    if r:
        raise VSError(r, "vs_ipc_open")
    return p.value


def vs_ipc_close(base_ptr: int):
    lib().vs_ipc_close(c_void_p(base_ptr))


class Runtime:
    """Owns one vs_rt handle; every method is a direct call of the C function of the same name."""

    def __init__(self, cfg: vs_config | None = None, **kw):
        L = lib()
        self.cfg = cfg if cfg is not None else vs_config_default(**kw)   # keeps the callbacks alive
        h = c_void_p()
        r = L.vs_create(ctypes.byref(self.cfg), ctypes.byref(h))
        if r:
            raise VSError(r, "vs_create")
        self.h = h
        self._keep = []   # ctypes callbacks kept alive

    def _ck(self, r, what=""):
        if r:
            raise VSError(r, (what + ": " if what else "") + self.vs_last_error())
        return r

    def vs_last_error(self) -> str:
        return lib().vs_last_error(self.h).decode()

    def vs_destroy(self):
        if self.h:
            lib().vs_destroy(self.h)
            self.h = None

    def close(self):
        self.vs_destroy()

    def __del__(self):
        try:
            self.vs_destroy()
        except Exception:
            pass

    def vs_type_create(self, name, modes):
        out = c_int32()
        m = (c_int * len(modes))(*modes)
        self._ck(lib().vs_type_create(self.h, name.encode(), len(modes), m, ctypes.byref(out)), "vs_type_create")
        return out.value

    def vs_version_add(self, ttype, name, gpu_mask, fn=None, user=None):
        """fn: a C function (a ctypes function of a loaded library, or its address as an int:
        called by the runtime directly, no Python in the loop), or a Python callable with the
        vs_launch_fn signature (called through a ctypes trampoline), or None (SIM only)."""
        if fn is None:
            cb = ctypes.cast(None, VS_LAUNCH_FN)
        elif isinstance(fn, int):
            cb = VS_LAUNCH_FN(fn)
        elif isinstance(fn, ctypes._CFuncPtr):
            cb = ctypes.cast(fn, VS_LAUNCH_FN)
        else:
            cb = VS_LAUNCH_FN(fn)
        self._keep.append(cb)
        out = c_int32()
        self._ck(lib().vs_version_add(self.h, ttype, name.encode(), gpu_mask, cb, user, ctypes.byref(out)),
                 "vs_version_add")
        return out.value

    def vs_register_builtins(self, dtype, version_mask):
        out = (c_int32 * VS_NUM_BUILTIN_TYPES)()
        self._ck(lib().vs_register_builtins(self.h, dtype, version_mask, out), "vs_register_builtins")
        return list(out)

    def vs_data_register(self, ptr, device, nbytes):
        out = c_int64()
        self._ck(lib().vs_data_register(self.h, c_void_p(ptr), device, nbytes, ctypes.byref(out)), "vs_data_register")
        return out.value

    def vs_submit(self, ttype, args, scalars: bytes | None = None):
        out = c_int64()
        a = _ids(args)
        sp = ctypes.c_char_p(scalars) if scalars else None
        self._ck(lib().vs_submit(self.h, ttype, a, len(args), ctypes.cast(sp, c_void_p) if sp else None,
                                 len(scalars) if scalars else 0, ctypes.byref(out)), "vs_submit")
        return out.value

    def vs_wait_all(self):
        return self._ck(lib().vs_wait_all(self.h), "vs_wait_all")

    def vs_wait_all_noflush(self):
        return self._ck(lib().vs_wait_all_noflush(self.h), "vs_wait_all_noflush")

    def vs_wait_on(self, d):
        return self._ck(lib().vs_wait_on(self.h, d), "vs_wait_on")

    def vs_stats(self) -> vs_stats_t:
        s = vs_stats_t()
        lib().vs_stats(self.h, ctypes.byref(s))
        return s

    def vs_group_stats(self):
        out = []
        for i in range(lib().vs_group_count(self.h)):
            g = vs_group_stat_t()
            lib().vs_group_stat(self.h, i, ctypes.byref(g))
            out.append({"type": g.type, "type_name": lib().vs_type_name(self.h, g.type).decode(),
                        "bytes": g.dataset_bytes, "reliable": bool(g.reliable),
                        "first_reliable": g.first_reliable_decision, "decisions": g.decisions,
                        "n": list(g.n[:g.nversions]), "mean_ns": list(g.mean_ns[:g.nversions]),
                        "assigned": list(g.assigned[:g.nversions]),
                        "versions": [lib().vs_version_name(self.h, g.type, v).decode() for v in range(g.nversions)]})
        return out

    def vs_decision_log(self):
        n = c_int64()
        lib().vs_decision_log(self.h, None, 0, ctypes.byref(n))
        buf = (vs_decision_t * max(1, n.value))()
        lib().vs_decision_log(self.h, buf, n.value, ctypes.byref(n))
        return [(r.task, r.version, r.worker, r.t_decide_ns, r.t_start_ns, r.t_end_ns, r.phase, r.type)
                for r in buf[:n.value]]

    def vs_decision_launches(self):
        """vs_decision_t.launch of every record (kernel launch number; grouped tasks share one)."""
        n = c_int64()
        lib().vs_decision_log(self.h, None, 0, ctypes.byref(n))
        buf = (vs_decision_t * max(1, n.value))()
        lib().vs_decision_log(self.h, buf, n.value, ctypes.byref(n))
        return [r.launch for r in buf[:n.value]]

    def vs_decision_issue_ns(self):
        n = c_int64()
        lib().vs_decision_issue_ns(self.h, None, 0, ctypes.byref(n))
        buf = (c_int64 * max(1, n.value))()
        lib().vs_decision_issue_ns(self.h, buf, n.value, ctypes.byref(n))
        return list(buf[:n.value])

    def vs_depend_on_event(self, event):
        """The next drive's device work waits for `event` (a torch.cuda.Event or a raw cudaEvent_t)."""
        h = getattr(event, "cuda_event", event)
        return self._ck(lib().vs_depend_on_event(self.h, c_void_p(int(h))), "vs_depend_on_event")

    def vs_transfer_plan(self):
        """Data ids of the batch's host-homed inputs in transfer order (vs_transfer_plan)."""
        n = c_int64()
        self._ck(lib().vs_transfer_plan(self.h, None, 0, ctypes.byref(n)), "vs_transfer_plan")
        buf = (c_int64 * max(1, n.value))()
        self._ck(lib().vs_transfer_plan(self.h, buf, n.value, ctypes.byref(n)), "vs_transfer_plan")
        return list(buf[:n.value])

    def vs_decision_log_hash(self) -> int:
        return int(lib().vs_decision_log_hash(self.h))

    def vs_decision_log_clear(self):
        return self._ck(lib().vs_decision_log_clear(self.h), "vs_decision_log_clear")

    def vs_table_dump(self, path):
        return self._ck(lib().vs_table_dump(self.h, path.encode()), "vs_table_dump")

    def vs_table_load(self, path):
        return self._ck(lib().vs_table_load(self.h, path.encode()), "vs_table_load")

    def vs_replay_set(self, ttype, nbytes, version, ns):
        return self._ck(lib().vs_replay_set(self.h, ttype, nbytes, version, ns), "vs_replay_set")

    def vs_data_invalidate(self, d):
        return self._ck(lib().vs_data_invalidate(self.h, d), "vs_data_invalidate")

    def vs_data_invalidate_n(self, ids):
        a = ids if isinstance(ids, ctypes.Array) else _ids(list(ids))
        return self._ck(lib().vs_data_invalidate_n(self.h, ctypes.cast(a, c_void_p), len(a)), "vs_data_invalidate_n")

    def vs_gpu_ordinal(self, g=0):
        r = lib().vs_gpu_ordinal(self.h, g)
        if r < 0:
            raise VSError(r, "vs_gpu_ordinal(%d)" % g)
        return r

    def vs_dist_init(self, rank, nranks, shm_name=""):
        return self._ck(lib().vs_dist_init(self.h, rank, nranks, shm_name.encode()), "vs_dist_init")

    def vs_data_set_owner(self, d, owner):
        return self._ck(lib().vs_data_set_owner(self.h, d, owner), "vs_data_set_owner")

    def vs_app_matmul(self, mm_type, m, l, n, A, B, C):
        return self._ck(lib().vs_app_matmul(self.h, mm_type, m, l, n, _ids(A), _ids(B), _ids(C)), "vs_app_matmul")

    def vs_app_cholesky(self, types, nt, A):
        """A: dict or list indexed i*nt+j (only i >= j used); missing entries may be -1."""
        arr = [-1] * (nt * nt)
        items = A.items() if isinstance(A, dict) else enumerate(A)
        for k, v in items:
            arr[k] = v
        return self._ck(lib().vs_app_cholesky(self.h, _ids(types, c_int32), nt, _ids(arr)), "vs_app_cholesky")
