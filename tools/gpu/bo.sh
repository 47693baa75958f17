CHOL_LIB_OVERRIDE=variants/phases.so python tools/phases_run.py factor 46080
CHOL_LIB_OVERRIDE=variants/phases_bo2k.so python tools/phases_run.py factor 46080
python tools/env_time.py 19200,46080 ""
CHOL_LIB_OVERRIDE=variants/bo2k.so python tools/env_time.py 9600,19200,46080 ""
