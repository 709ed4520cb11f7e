#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build94.log 2>&1
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/t94.log 2>&1; echo "exit $?" >> gpurun_out/t94.log
timeout 300 python __graft_entry__.py smoke > gpurun_out/smoke94.log 2>&1; echo "exit $?" >> gpurun_out/smoke94.log
