#!/bin/bash
# edge-case tests (b=4096 sampled rows, unsupported sizes, empty / one-tile graphs)
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_tiles.py tests/test_gpu_runtime.py -q -p no:cacheprovider -k "4096 or unsupported or empty" > gpurun_out/t81.log 2>&1; echo "exit $?" >> gpurun_out/t81.log
