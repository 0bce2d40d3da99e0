cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
O=gpurun_out/diag8.log; : > $O
run() { echo "== $*" >> $O; timeout 100 env "$@" >> $O 2>&1 || echo "rc=$?" >> $O; }
run DIAG_TIMEOUT=60 python tools/split_diag.py C2 0 5
run DIAG_TIMEOUT=60 CULI_STEAL_GATE=0 python tools/split_diag.py C2 0 5
run DIAG_TIMEOUT=60 CULI_SPLIT_POLL=128 python tools/split_diag.py C2 0 5
run DIAG_TIMEOUT=60 CULI_SPLIT_POLL=32 python tools/split_diag.py C2 0 5
run DIAG_TIMEOUT=60 CULI_SPLIT_SLEEP=1024 python tools/split_diag.py C2 0 5
run DIAG_TIMEOUT=60 python tools/split_diag.py C5 0 5
run DIAG_TIMEOUT=60 CULI_STEAL_GATE=0 python tools/split_diag.py C5 0 5
run DIAG_TIMEOUT=60 DIAG_N=5000 python tools/split_diag.py C5 1 10
grep -v "Exception ignored\|culi.py\", line 28\|NoneType\|^Traceback" $O
