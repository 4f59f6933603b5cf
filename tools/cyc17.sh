#!/bin/bash
# locate the GPU-suite crash; host partition timing plain vs write-combining
mkdir -p gpurun_out
for f in tests/test_gpu_*.py; do echo "== $f"; timeout 900 python -X faulthandler -m pytest $f -m gpu -x -q 2>&1 | grep -E "passed|failed|error|Fatal|File \"/root|line [0-9]+ in test" | head -8; done
python - <<'PY'
import torch, time
from paper_conf_cidr_chrysogelossa19_b200 import host_partition
import os
k=torch.randint(-2**31,2**31,(1<<27,),dtype=torch.int32); p=torch.randint(-2**31,2**31,(1<<27,),dtype=torch.int32)
for i in range(3):
    t=time.time(); host_partition(k,p,3); print("plain 2^27 int32 F=8:", round(time.time()-t,3), flush=True)
PY
HAPE_HP_WC=1 python - <<'PY'
import torch, time
from paper_conf_cidr_chrysogelossa19_b200 import host_partition
k=torch.randint(-2**31,2**31,(1<<27,),dtype=torch.int32); p=torch.randint(-2**31,2**31,(1<<27,),dtype=torch.int32)
for i in range(3):
    t=time.time(); host_partition(k,p,3); print("wc 2^27 int32 F=8:", round(time.time()-t,3), flush=True)
for T in (4, 8, 16):
    t=time.time(); host_partition(k,p,3, threads=T); print("wc T", T, round(time.time()-t,3), flush=True)
PY
