#!/bin/bash
# warm-start cold step: lazy vs eager module loading
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 400 python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --table-dump gpurun_out/table96.json > gpurun_out/b96_dump.log 2>&1
timeout 400 python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --table-load gpurun_out/table96.json > gpurun_out/b96_load_lazy.log 2>&1
CUDA_MODULE_LOADING=EAGER timeout 400 python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --table-load gpurun_out/table96.json > gpurun_out/b96_load_eager.log 2>&1
